#!/usr/bin/env python
"""Per-instruction stall reasons from an ncu report: the dispatch-stalled / wait-stalled instructions,
and a window of SASS around the hottest loop.

    python tools/ncu_stalls.py report.ncu-rep [reason] [--top N] [--range A B]
"""
import csv
import io
import subprocess
import sys


def load(rep):
    if rep.endswith(".gz"):
        import gzip
        out = gzip.open(rep, "rt").read()
    elif rep.endswith(".csv"):
        out = open(rep).read()
    else:
        out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                             capture_output=True, text=True).stdout
    lines = out.splitlines()
    rd = csv.reader(io.StringIO("\n".join(lines[1:])))
    hdr = next(rd)
    return hdr, [r for r in rd if len(r) == len(hdr)]


def main():
    rep = sys.argv[1]
    reason = sys.argv[2] if len(sys.argv) > 2 and not sys.argv[2].startswith("--") else "stall_dispatch"
    top = int(sys.argv[sys.argv.index("--top") + 1]) if "--top" in sys.argv else 30
    hdr, rows = load(rep)
    ir = hdr.index(reason)
    isrc = hdr.index("Source")
    iad = hdr.index("Address")
    iex = hdr.index("Instructions Executed")
    if "--range" in sys.argv:
        a = int(sys.argv[sys.argv.index("--range") + 1])
        b = int(sys.argv[sys.argv.index("--range") + 2])
        cols = [hdr.index(c) for c in ("stall_selected", "stall_not_selected", "stall_dispatch", "stall_wait",
                                       "stall_short_sb", "stall_branch_resolving", "stall_no_inst")]
        print("idx   exec  sel  nsel disp wait ssb  br  noi  sass")
        for i in range(a, min(b, len(rows))):
            r = rows[i]
            print(f"{i:5d} {int(r[iex] or 0) // 1000:6d}k " + " ".join(f"{int(r[c] or 0):4d}" for c in cols) +
                  "  " + r[isrc].strip())
        return
    order = sorted(range(len(rows)), key=lambda i: -int(rows[i][ir] or 0))[:top]
    tot = sum(int(r[ir] or 0) for r in rows)
    print(f"{reason}: total samples {tot}")
    for i in order:
        r = rows[i]
        print(f"{i:5d} {int(r[ir] or 0):6d}  {r[isrc].strip()}")


if __name__ == "__main__":
    main()

#!/usr/bin/env python
"""Dynamic SASS instruction mix and stall samples per opcode from an ncu report's source page.

    python tools/ncu_sass_mix.py report.ncu-rep [--top N]
"""
import collections
import csv
import io
import re
import subprocess
import sys


def main():
    rep = sys.argv[1]
    top = int(sys.argv[sys.argv.index("--top") + 1]) if "--top" in sys.argv else 0
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
    iex = hdr.index("Instructions Executed")
    ist = hdr.index("Warp Stall Sampling (All Samples)")
    isrc = hdr.index("Source")
    mix = collections.Counter()
    stall = collections.Counter()
    rows = []
    for r in rd:
        if len(r) <= iex:
            continue
        src = r[isrc].strip()
        op = re.sub(r"^@!?U?P\w+\s+", "", src).split(" ")[0].split(".")[0]
        n = int(r[iex] or 0)
        s = int(r[ist] or 0)
        mix[op] += n
        stall[op] += s
        rows.append((s, n, src))
    tot = sum(mix.values())
    stot = sum(stall.values())
    print(f"executed warp-instructions: {tot}")
    for op, n in mix.most_common(25):
        print(f"  {op:14s} {n:12d} {100 * n / tot:6.2f}%   stall-samples {100 * stall[op] / max(stot, 1):5.1f}%")
    if top:
        for s, n, src in sorted(rows, reverse=True)[:top]:
            print(f"  {s:7d} {n:10d}  {src}")


if __name__ == "__main__":
    main()

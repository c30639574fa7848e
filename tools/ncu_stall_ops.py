#!/usr/bin/env python
"""Stall samples per opcode and per reason from an ncu source-page CSV (.csv or .csv.gz), plus the
instructions carrying the most samples of one reason.

    python tools/ncu_stall_ops.py X.src.csv.gz [--reason stall_wait] [--top 15]
"""
import collections
import csv
import gzip
import io
import re
import sys


def main():
    path = sys.argv[1]
    reason = sys.argv[sys.argv.index("--reason") + 1] if "--reason" in sys.argv else "stall_wait"
    top = int(sys.argv[sys.argv.index("--top") + 1]) if "--top" in sys.argv else 15
    text = gzip.open(path, "rt").read() if path.endswith(".gz") else open(path).read()
    rd = csv.reader(io.StringIO("\n".join(text.splitlines()[1:])))
    hdr = next(rd)
    reasons = [h for h in hdr if h.startswith("stall_") and "Not Issued" not in h]
    idx = {h: hdr.index(h) for h in reasons}
    iex = hdr.index("Instructions Executed")
    per_op = collections.defaultdict(collections.Counter)
    rows = []
    for r in rd:
        if len(r) <= iex:
            continue
        op = re.sub(r"^@!?U?P\w+\s+", "", r[1].strip()).split(" ")[0].split(".")[0]
        for h in reasons:
            v = int(r[idx[h]] or 0)
            per_op[op][h] += v
        rows.append((int(r[idx[reason]] or 0), r[1].strip()[:70], r[iex]))
    tot = sum(sum(c.values()) for c in per_op.values())
    print(f"total samples {tot}")
    for op, c in sorted(per_op.items(), key=lambda kv: -sum(kv[1].values()))[:12]:
        s = sum(c.values())
        top3 = ", ".join(f"{h[6:]} {100 * v / tot:.1f}" for h, v in c.most_common(4) if v)
        print(f"{op:10s} {100 * s / tot:5.1f}%  {top3}")
    print(f"-- top {reason}:")
    for v, src, n in sorted(rows, reverse=True)[:top]:
        print(f"{100 * v / tot:5.2f}%  {src}  (exec {n})")


if __name__ == "__main__":
    main()

#!/usr/bin/env python
"""SASS evidence for a kernel of libconv2d.so: opcode histogram, LDL/STL (spill) count, FFMA share.

    python tools/sass_stats.py <function-name-regex> [--dump]
"""
import collections
import os
import re
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
LIB = os.path.join(ROOT, "paper_conf_cluster_luzw20_b200", "libconv2d.so")


def functions(lib=LIB):
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "-sass", lib], capture_output=True, text=True).stdout
    funcs, cur = {}, None
    for ln in out.splitlines():
        m = re.search(r"Function : (\S+)", ln)
        if m:
            cur = m.group(1)
            funcs[cur] = []
        elif cur:
            funcs[cur].append(ln)
    return funcs


def opcodes(lines):
    ops = []
    for ln in lines:
        m = re.match(r"\s+/\*[0-9a-f]{4,}\*/\s+(@!?U?P\w+\s+)?([A-Z][A-Z0-9_.]+)", ln)
        if m:
            ops.append(m.group(2))
    return ops


def main():
    pat = re.compile(sys.argv[1])
    for name, lines in functions().items():
        if not pat.search(name):
            continue
        ops = opcodes(lines)
        base = collections.Counter(o.split(".")[0] for o in ops)
        print(f"== {name}: {len(ops)} instructions, FFMA {base['FFMA']} ({100 * base['FFMA'] / max(1, len(ops)):.1f}%), "
              f"LDL {base['LDL']} STL {base['STL']}")
        print("   " + ", ".join(f"{k} {v}" for k, v in base.most_common(25)))
        if "--dump" in sys.argv:
            print("\n".join(lines))


if __name__ == "__main__":
    main()

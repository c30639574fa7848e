#!/usr/bin/env python
"""SASS evidence of the built libraries (north_star: "committed ncu and SASS evidence").

    python tools/sass_report.py [--lib product|tune] [--out profiles/<tag>_sass_product.txt]

For every kernel of the library: instruction count and the opcode histogram that carries the paper's
claims on sm_100a -- FFMA (the row-reuse FMAs), SHFL (column reuse), FSEL/SEL (Alg. 1's select),
LDCU/LDC (uniform-register filter operands), LDS (shared-memory filter / row ring), LDG/LDGSTS
(row fetch), STG (output rows), LDL/STL (register spills: must be 0), and the tcgen05 / TMA opcodes
(UTCHMMA / UTCQMMA, LDTM, STTM, UBLKCP) of the tensor-core variant. Plus the ptxas register / spill
table (-Xptxas -v of every unit, product flags).
"""
import argparse
import collections
import os
import re
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PKG = os.path.join(ROOT, "paper_conf_cluster_luzw20_b200")
LIBS = {"product": os.path.join(PKG, "libconv2d.so"), "tune": os.path.join(PKG, "libconv2d_tune.so")}
COLS = ["FFMA", "FFMA2", "SHFL", "FSEL", "SEL", "LDCU", "LDC", "LDS", "LDG", "LDGSTS", "STG", "STS", "LDL", "STL",
        "UTCHMMA", "UTCQMMA", "LDTM", "STTM", "UBLKCP", "BAR", "SYNCS"]


def kernels(lib):
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "-sass", lib], capture_output=True, text=True,
                         check=True).stdout
    res, cur = {}, None
    for ln in out.splitlines():
        m = re.search(r"Function : (\S+)", ln)
        if m:
            cur = m.group(1)
            res[cur] = collections.Counter()
            continue
        if cur is None:
            continue
        m = re.match(r"\s+/\*[0-9a-f]{4,}\*/\s+(@!?U?P\w+\s+)?([A-Z][A-Z0-9_.]+)", ln)
        if m:
            res[cur][m.group(2).split(".")[0]] += 1
    return res


def demangle(names):
    r = subprocess.run(["c++filt"], input="\n".join(names), capture_output=True, text=True)
    return r.stdout.splitlines() if r.returncode == 0 else list(names)


def spills(lib):
    """{kernel: (LDL, STL)} for every kernel with local-memory traffic."""
    return {k: (c["LDL"], c["STL"]) for k, c in kernels(lib).items() if c["LDL"] or c["STL"]}


def ptxas_table():
    sys.path.insert(0, ROOT)
    from paper_conf_cluster_luzw20_b200 import _build

    rows = []
    for src in _build.sources():
        cmd = [_build.NVCC, *_build.ARCH, *_build.FLAGS, "-I", os.path.join(ROOT, "include"), "-Xptxas=-v", "-c",
               "-o", "/dev/null", src]
        err = subprocess.run(cmd, capture_output=True, text=True).stderr
        cur = None
        for ln in err.splitlines():
            m = re.search(r"Compiling entry function '(\S+)'", ln)
            if m:
                cur = m.group(1)
            m = re.search(r"(\d+) bytes stack frame, (\d+) bytes spill stores, (\d+) bytes spill loads", ln)
            if m and cur:
                rows.append([cur, None, int(m.group(2)), int(m.group(3))])
            m = re.search(r"Used (\d+) registers", ln)
            if m and rows and rows[-1][0] == cur and rows[-1][1] is None:
                rows[-1][1] = int(m.group(1))
    return rows


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--lib", default="product", choices=sorted(LIBS))
    ap.add_argument("--out", default=None)
    ap.add_argument("--no-ptxas", action="store_true")
    a = ap.parse_args()
    ks = kernels(LIBS[a.lib])
    names = sorted(ks)
    pretty = dict(zip(names, demangle(names)))
    lines = [f"# SASS opcode histogram of {os.path.basename(LIBS[a.lib])} ({len(ks)} kernels; cuobjdump -sass)",
             "# kernel | total | " + " ".join(COLS)]
    for k in names:
        c = ks[k]
        lines.append(f"{pretty[k]} | {sum(c.values())} | " + " ".join(f"{col}={c[col]}" for col in COLS if c[col]))
    sp = {k: (c["LDL"], c["STL"]) for k, c in ks.items() if c["LDL"] or c["STL"]}
    lines.append(f"# kernels with LDL/STL (spills): {len(sp)}")
    for k, v in sorted(sp.items()):
        lines.append(f"#   {pretty[k]}: LDL {v[0]} STL {v[1]}")
    if not a.no_ptxas and a.lib == "product":
        lines.append("# ptxas -v (product flags): kernel | registers | spill stores | spill loads (bytes)")
        rows = ptxas_table()
        pr = dict(zip([r[0] for r in rows], demangle([r[0] for r in rows])))
        for r in rows:
            lines.append(f"{pr[r[0]]} | {r[1]} | {r[2]} | {r[3]}")
    text = "\n".join(lines) + "\n"
    if a.out:
        with open(a.out, "w") as fh:
            fh.write(text)
    sys.stdout.write(text if not a.out else f"wrote {a.out}: {len(ks)} kernels, {len(sp)} with spills\n")


if __name__ == "__main__":
    main()

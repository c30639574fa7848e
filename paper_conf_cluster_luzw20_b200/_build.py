"""Build libconv2d.so (the C-ABI library) in-tree for sm_100a with nvcc, and its tuning twin
libconv2d_tune.so (same sources with -DC2D_TUNING: every kernel variant instantiated and the
c2d_debug_set_* switches exported, for tools/ and the variant-equivalence tests; the product library
has the tuned defaults only).

    python -m paper_conf_cluster_luzw20_b200._build [--force] [--verbose] [--product-only]

Flags: -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo, no fast-math (fp32 FMA contraction is
allowed, denormals preserved: DESIGN.md R5). Static cudart, so the .so only needs the driver.
Every csrc/*.cu is one translation unit (one per K plus the C-ABI unit), compiled in parallel to an
object in build/ and linked into the shared library.
"""
from __future__ import annotations

import concurrent.futures
import glob
import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
LIB = os.path.join(PKG, "libconv2d.so")
LIB_TUNE = os.path.join(PKG, "libconv2d_tune.so")
HEADER = os.path.join(ROOT, "include", "conv2d.h")

NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
FLAGS = ["-O3", "-lineinfo", "-std=c++17", "-Xcompiler", "-fPIC", "--ftz=false", "--prec-div=true",
         "--prec-sqrt=true", "--fmad=true"]
OBJDIR = os.path.join(ROOT, "build", "csrc_obj")
OBJDIR_TUNE = os.path.join(ROOT, "build", "csrc_obj_tune")


def sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")))


def _stale(lib: str) -> bool:
    if not os.path.exists(lib):
        return True
    t = os.path.getmtime(lib)
    deps = sources() + glob.glob(os.path.join(CSRC, "*.cuh")) + glob.glob(os.path.join(CSRC, "*.h")) + [HEADER, __file__]
    return any(os.path.getmtime(d) > t for d in deps)


def _compile(src: str, objdir: str, defines: list, verbose: bool) -> str:
    obj = os.path.join(objdir, os.path.basename(src).replace(".cu", ".o"))
    cmd = [NVCC, *ARCH, *FLAGS, *defines, "-I", os.path.join(ROOT, "include"), "-c", "-o", obj, src]
    if verbose:
        cmd.insert(1, "-Xptxas=-v")
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"nvcc failed ({' '.join(cmd)}):\n{r.stdout}\n{r.stderr}")
    if verbose:
        sys.stderr.write(r.stderr)
    return obj


def _link(objs: list, lib: str) -> None:
    tmp = lib + f".tmp{os.getpid()}"
    cmd = [NVCC, *ARCH, "-shared", "-cudart", "static", "-o", tmp, *objs]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"link failed ({' '.join(cmd)}):\n{r.stdout}\n{r.stderr}")
    os.replace(tmp, lib)


def build(force: bool = False, verbose: bool = False, jobs: int = 0, tuning: bool = True) -> str:
    """Build the product library (and, unless tuning=False, the tuning library); returns LIB."""
    targets = [(LIB, OBJDIR, [])]
    if tuning:
        targets.append((LIB_TUNE, OBJDIR_TUNE, ["-DC2D_TUNING"]))
    targets = [t for t in targets if force or _stale(t[0])]
    if not targets:
        return LIB
    for _, objdir, _ in targets:
        os.makedirs(objdir, exist_ok=True)
    work = [(src, objdir, defs) for _, objdir, defs in targets for src in sources()]
    # the largest units (the per-K kernel units, K = 15 first) go first
    work.sort(key=lambda w: -os.path.getsize(w[0]) - (int(w[0][-5:-3]) if w[0][-5:-3].isdigit() else 0) * 1000)
    jobs = jobs or max(1, os.cpu_count() or 1)
    with concurrent.futures.ThreadPoolExecutor(jobs) as ex:
        objs = list(ex.map(lambda w: _compile(w[0], w[1], w[2], verbose), work))
    for lib, objdir, _ in targets:
        _link([o for o in objs if os.path.dirname(o) == objdir], lib)
    return LIB


if __name__ == "__main__":
    print(build(force="--force" in sys.argv, verbose="--verbose" in sys.argv,
                tuning="--product-only" not in sys.argv))

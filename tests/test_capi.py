"""CPU-side checks of the boundary: libconv2d.so builds for sm_100a, loads, and exports every symbol
include/conv2d.h declares; the binding mirrors the header; host-side argument errors are reported
without touching a GPU. No compute calls (no GPU here)."""
import ctypes
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "conv2d.h")


@pytest.fixture(scope="module")
def lib():
    from paper_conf_cluster_luzw20_b200 import _build, _capi

    _build.build()
    return _capi.load()


def _declared_functions():
    text = open(HEADER).read()
    text = re.sub(r"/\*.*?\*/", "", text, flags=re.S)
    return sorted(set(re.findall(r"^\s*(?:const\s+)?\w+\s*\*?\s*(conv2d_\w+)\s*\(", text, flags=re.M)))


def test_header_declares_the_boundary():
    funcs = _declared_functions()
    for f in ("conv2d_single", "conv2d_multi", "conv2d_strerror"):
        assert f in funcs


def test_every_declared_symbol_is_exported(lib):
    from paper_conf_cluster_luzw20_b200 import _capi

    funcs = _declared_functions()
    assert sorted(funcs) == sorted(_capi.EXPORTS)
    for f in funcs:
        assert hasattr(lib, f), f
    out = subprocess.run(["nm", "-D", "--defined-only", _capi.LIB_PATH], capture_output=True, text=True).stdout
    for f in funcs:
        assert re.search(rf"\bT {f}$", out, flags=re.M), f"{f} not exported with C linkage"


def test_error_codes_match_header(lib):
    from paper_conf_cluster_luzw20_b200 import _capi

    text = open(HEADER).read()
    codes = {m[0]: int(m[1]) for m in re.findall(r"#define (CONV2D_\w+) \(?(-?\d+)\)?", text)}
    assert codes["CONV2D_OK"] == _capi.CONV2D_OK
    assert codes["CONV2D_ENULL"] == _capi.CONV2D_ENULL
    assert codes["CONV2D_ESHAPE"] == _capi.CONV2D_ESHAPE
    assert codes["CONV2D_EK"] == _capi.CONV2D_EK
    assert codes["CONV2D_EOVERLAP"] == _capi.CONV2D_EOVERLAP
    assert codes["CONV2D_ECUDA"] == _capi.CONV2D_ECUDA
    assert codes["CONV2D_EALIGN"] == _capi.CONV2D_EALIGN
    assert codes["CONV2D_MAX_K"] == _capi.CONV2D_MAX_K
    for c in codes.values():
        assert isinstance(_capi.strerror(c), str) and _capi.strerror(c)
    assert lib.conv2d_version() >= 100


def test_argument_errors_need_no_gpu(lib):
    """Validation happens before any CUDA call: these return their codes on a GPU-less host."""
    from paper_conf_cluster_luzw20_b200 import _capi as c

    a, b, o = 0x10000, 0x20000000, 0x40000000  # fake, never dereferenced
    assert c.conv2d_single(None, 8, 8, b, 3, o) == c.CONV2D_ENULL
    assert c.conv2d_single(a, 8, 8, None, 3, o) == c.CONV2D_ENULL
    assert c.conv2d_single(a, 8, 8, b, 16, o) == c.CONV2D_EK
    assert c.conv2d_single(a, 8, 8, b, 0, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single(a, 2, 8, b, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single(a, 8, 2, b, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single(a + 2, 8, 8, b, 3, o) == c.CONV2D_EALIGN
    assert c.conv2d_single(a, 8, 8, b, 3, a + 16) == c.CONV2D_EOVERLAP
    assert c.conv2d_single(a, 8, 8, b, 3, b) == c.CONV2D_EOVERLAP
    assert c.conv2d_multi(a, 0, 1, 8, 8, b, 1, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_multi(a, 1, 0, 8, 8, b, 1, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_multi(a, 1, 1, 8, 8, b, 0, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_multi(a, 1, 1, 8, 8, b, 1, 16, o) == c.CONV2D_EK
    assert c.conv2d_multi(a, 2, 2, 8, 8, b, 1, 3, a + 100) == c.CONV2D_EOVERLAP
    assert c.conv2d_single_direct(a, 8, 8, b, 20, o) == c.CONV2D_EK
    # conv2d_single_halo (N3): rows of `in` then rows of `halo`
    h = 0x60000000
    assert c.conv2d_single_halo(a, 8, 8, None, 2, b, 3, o) == c.CONV2D_ENULL
    assert c.conv2d_single_halo(a, 8, 8, h, -1, b, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single_halo(a, 8, 8, h, 2, b, 16, o) == c.CONV2D_EK
    assert c.conv2d_single_halo(a, 1, 8, h, 1, b, 3, o) == c.CONV2D_ESHAPE  # 2 rows < K
    assert c.conv2d_single_halo(a, 8, 8, h + 2, 2, b, 3, o) == c.CONV2D_EALIGN
    assert c.conv2d_single_halo(a, 8, 8, h, 2, b, 3, h + 8) == c.CONV2D_EOVERLAP
    # conv2d_single_pad (N4): mode bits, 'same' allows images smaller than the filter
    assert c.conv2d_single_pad(a, 8, 8, b, 3, 3, o) == c.CONV2D_ESHAPE  # both PAD flags
    assert c.conv2d_single_pad(a, 8, 8, b, 3, 8, o) == c.CONV2D_ESHAPE  # unknown bit
    assert c.conv2d_single_pad(None, 8, 8, b, 3, 1, o) == c.CONV2D_ENULL
    assert c.conv2d_single_pad(a, 8, 8, b, 16, 1, o) == c.CONV2D_EK
    assert c.conv2d_single_pad(a, 2, 8, b, 3, c.CONV2D_FLIP, o) == c.CONV2D_ESHAPE  # valid needs H >= K
    assert c.conv2d_single_pad(a, 0, 8, b, 3, 1, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single_pad(a, 8, 8, b, 3, 2, a + 32) == c.CONV2D_EOVERLAP


def test_library_is_sm100a(lib):
    from paper_conf_cluster_luzw20_b200 import _capi

    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", _capi.LIB_PATH],
                         capture_output=True, text=True).stdout
    assert "sm_100a" in out


def test_product_path_has_no_oracle_dependency():
    """The package never imports or links the oracle (they share no code)."""
    pkg = os.path.join(ROOT, "paper_conf_cluster_luzw20_b200")
    for dirpath, _, files in os.walk(pkg):
        for fn in files:
            if fn.endswith((".py", ".cu", ".cuh", ".h", ".c", ".cpp")):
                src = open(os.path.join(dirpath, fn)).read()
                assert "import oracle" not in src and "from oracle" not in src, fn
                assert "liboracle" not in src and "conv2d_oracle" not in src, fn


def test_batch_argument_errors_need_no_gpu(lib):
    from paper_conf_cluster_luzw20_b200 import _capi as c

    a, b, o = 0x10000, 0x20000000, 0x40000000  # fake, never dereferenced
    assert c.conv2d_single_batch(None, 2, 8, 8, b, 3, o) == c.CONV2D_ENULL
    assert c.conv2d_single_batch(a, 0, 8, 8, b, 3, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single_batch(a, 2, 8, 8, b, 16, o) == c.CONV2D_EK
    assert c.conv2d_single_batch(a, 2, 2, 8, b, 3, o) == c.CONV2D_ESHAPE
    # the second image's input (bytes 256..512) overlaps the output
    assert c.conv2d_single_batch(a, 2, 8, 8, b, 3, a + 300) == c.CONV2D_EOVERLAP
    assert c.conv2d_multi_tc(a, 2, 2, 8, 8, b, 1, 3, a + 100) == c.CONV2D_EOVERLAP
    # conv2d_single_rect (N4): FH x FW in [1, 15]
    assert c.conv2d_single_rect(None, 8, 8, b, 3, 5, o) == c.CONV2D_ENULL
    assert c.conv2d_single_rect(a, 8, 8, b, 3, 16, o) == c.CONV2D_EK
    assert c.conv2d_single_rect(a, 8, 8, b, 0, 5, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single_rect(a, 8, 4, b, 3, 5, o) == c.CONV2D_ESHAPE
    assert c.conv2d_single_rect(a, 8, 8, b, 3, 5, a + 16) == c.CONV2D_EOVERLAP


def test_product_library_has_no_tuning_switches(lib):
    """The shipped libconv2d.so exports exactly the header's C ABI (no process-global tuning
    switches); the c2d_debug_set_* switches live in the separate tuning build libconv2d_tune.so."""
    from paper_conf_cluster_luzw20_b200 import _capi

    out = subprocess.run(["nm", "-D", "--defined-only", _capi.LIB_PATH], capture_output=True, text=True).stdout
    exported = set(re.findall(r"\bT (\w+)$", out, flags=re.M))
    c_linkage = {e for e in exported if not e.startswith("_Z")}  # C++ symbols are not the C ABI
    assert c_linkage == set(_capi.EXPORTS), c_linkage ^ set(_capi.EXPORTS)
    assert not any("debug" in e for e in exported)
    out = subprocess.run(["nm", "-D", "--defined-only", _capi.TUNE_LIB_PATH], capture_output=True, text=True).stdout
    for f in ("c2d_debug_set_variant", "c2d_debug_set_multi_variant", "c2d_debug_set_min_band"):
        assert re.search(rf"\bT {f}$", out, flags=re.M), f

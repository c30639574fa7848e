"""ctypes binding of libconv2d.so -- the C ABI of include/conv2d.h, same names, argument marshalling
only. Loading fails loudly if the library is missing (there is no CPU or PyTorch fallback).

`load_tuning()` loads the tuning twin libconv2d_tune.so (every kernel variant, c2d_debug_set_*
switches) for tools/ and the variant-equivalence tests; the product path never uses it."""
from __future__ import annotations

import ctypes
import os

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "libconv2d.so")
TUNE_LIB_PATH = os.path.join(_PKG, "libconv2d_tune.so")

# every symbol include/conv2d.h declares
EXPORTS = ("conv2d_single", "conv2d_single_batch", "conv2d_single_rect", "conv2d_multi", "conv2d_single_ex", "conv2d_multi_ex", "conv2d_single_halo",
           "conv2d_single_pad",
           "conv2d_single_direct",
           "conv2d_single_host", "conv2d_multi_tc", "conv2d_release_scratch", "conv2d_strerror", "conv2d_version")

CONV2D_OK = 0
CONV2D_ENULL = -1
CONV2D_ESHAPE = -2
CONV2D_EK = -3
CONV2D_EOVERLAP = -4
CONV2D_ECUDA = -5
CONV2D_EALIGN = -6
CONV2D_EALLOC = -7
CONV2D_MAX_K = 15
CONV2D_PAD_ZERO = 1
CONV2D_PAD_REPLICATE = 2
CONV2D_FLIP = 4

_lib = None
_tune = None


class Conv2dError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"{msg} (code {code})")
        self.code = code


def _declare(L):
    P, I = ctypes.c_void_p, ctypes.c_int
    L.conv2d_single.argtypes = [P, I, I, P, I, P, P]
    L.conv2d_single_ex.argtypes = [P, I, I, P, I, P, P, I]
    L.conv2d_single_batch.argtypes = [P, I, I, I, P, I, P, P]
    L.conv2d_single_rect.argtypes = [P, I, I, P, I, I, P, P]
    L.conv2d_single_halo.argtypes = [P, I, I, P, I, P, I, P, P]
    L.conv2d_single_pad.argtypes = [P, I, I, P, I, I, P, P]
    L.conv2d_single_direct.argtypes = [P, I, I, P, I, P, P]
    L.conv2d_multi.argtypes = [P, I, I, I, I, P, I, I, P, P]
    L.conv2d_multi_ex.argtypes = [P, I, I, I, I, P, I, I, P, P, I]
    L.conv2d_single_host.argtypes = [P, I, I, P, I, P, P, I]
    L.conv2d_multi_tc.argtypes = [P, I, I, I, I, P, I, I, P, P]
    L.conv2d_release_scratch.argtypes = []
    for f in EXPORTS:
        if f != "conv2d_strerror":
            getattr(L, f).restype = I
    L.conv2d_strerror.argtypes = [I]
    L.conv2d_strerror.restype = ctypes.c_char_p
    return L


def load(path: str | None = None):
    """Load libconv2d.so (built in-tree by __graft_entry__.build()). Raises if it is missing."""
    global _lib
    if _lib is not None:
        return _lib
    p = path or LIB_PATH
    if not os.path.exists(p):
        raise ImportError(f"{p} is missing: run `python -c 'import __graft_entry__ as g; g.build()'` "
                          "(there is no fallback implementation)")
    _lib = _declare(ctypes.CDLL(p))
    return _lib


def load_tuning():
    """The tuning library libconv2d_tune.so (tools/, variant tests): same C ABI plus the
    c2d_debug_set_* switches; a separate handle, the product library stays loaded as is."""
    global _tune
    if _tune is not None:
        return _tune
    if not os.path.exists(TUNE_LIB_PATH):
        raise ImportError(f"{TUNE_LIB_PATH} is missing: run `python -m paper_conf_cluster_luzw20_b200._build`")
    L = _declare(ctypes.CDLL(TUNE_LIB_PATH))
    for f in ("c2d_debug_set_variant", "c2d_debug_set_min_band", "c2d_debug_set_multi_variant"):
        getattr(L, f).argtypes = [ctypes.c_int]
        getattr(L, f).restype = ctypes.c_int
    _tune = L
    return L


_active = None  # the library the entry points below call: the product library unless switched


def lib():
    """The library the entry points call (hot path: one global lookup): libconv2d.so, or the tuning
    library after use_tuning_library() (tools/ and the variant tests only)."""
    if _active is not None:
        return _active
    return _lib if _lib is not None else load()


def use_tuning_library(on: bool = True) -> None:
    """Route every entry point of this module (and so of api.py) to libconv2d_tune.so (on=True) or
    back to the product libconv2d.so. For tuning tools and the variant-equivalence tests."""
    global _active
    _active = load_tuning() if on else None


class tuning_session:
    """`with tuning_session(variant=v):` -- entry points call the tuning library with variant v
    (multi_variant / min_band likewise), restored on exit."""

    def __init__(self, variant: int = 0, multi_variant: int = 0, min_band: int = 0):
        self.v, self.mv, self.mb = variant, multi_variant, min_band

    def __enter__(self):
        global _active
        self.prev = _active
        L = load_tuning()
        L.c2d_debug_set_variant(self.v)
        L.c2d_debug_set_multi_variant(self.mv)
        L.c2d_debug_set_min_band(self.mb)
        _active = L
        return L

    def __exit__(self, *exc):
        global _active
        L = load_tuning()
        L.c2d_debug_set_variant(0)
        L.c2d_debug_set_multi_variant(0)
        L.c2d_debug_set_min_band(0)
        _active = self.prev


def strerror(code: int) -> str:
    return lib().conv2d_strerror(int(code)).decode()


def check(code: int) -> None:
    if code != CONV2D_OK:
        raise Conv2dError(code, strerror(code))


# raw entry points (device pointers as ints, stream handle as int): same names as the C ABI
def conv2d_single(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0) -> int:
    return lib().conv2d_single(in_ptr, H, W, filt_ptr, K, out_ptr, stream)


def conv2d_single_batch(in_ptr, N, H, W, filt_ptr, K, out_ptr, stream=0) -> int:
    return lib().conv2d_single_batch(in_ptr, N, H, W, filt_ptr, K, out_ptr, stream)


def conv2d_single_rect(in_ptr, H, W, filt_ptr, FH, FW, out_ptr, stream=0) -> int:
    return lib().conv2d_single_rect(in_ptr, H, W, filt_ptr, FH, FW, out_ptr, stream)


def conv2d_single_ex(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0, band_h=0) -> int:
    return lib().conv2d_single_ex(in_ptr, H, W, filt_ptr, K, out_ptr, stream, band_h)


def conv2d_single_pad(in_ptr, H, W, filt_ptr, K, mode, out_ptr, stream=0) -> int:
    return lib().conv2d_single_pad(in_ptr, H, W, filt_ptr, K, mode, out_ptr, stream)


def conv2d_single_halo(in_ptr, H, W, halo_ptr, halo_rows, filt_ptr, K, out_ptr, stream=0) -> int:
    return lib().conv2d_single_halo(in_ptr, H, W, halo_ptr, halo_rows, filt_ptr, K, out_ptr, stream)


def conv2d_single_direct(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0) -> int:
    return lib().conv2d_single_direct(in_ptr, H, W, filt_ptr, K, out_ptr, stream)


def conv2d_multi(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream=0) -> int:
    return lib().conv2d_multi(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream)


def conv2d_multi_ex(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream=0, band_h=0) -> int:
    return lib().conv2d_multi_ex(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream, band_h)


def conv2d_single_host(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0, chunk_rows=0) -> int:
    return lib().conv2d_single_host(in_ptr, H, W, filt_ptr, K, out_ptr, stream, chunk_rows)


def conv2d_multi_tc(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream=0) -> int:
    return lib().conv2d_multi_tc(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream)


def conv2d_release_scratch() -> int:
    return lib().conv2d_release_scratch()


def conv2d_version() -> int:
    return lib().conv2d_version()


_switches = {"variant": 0, "multi_variant": 0, "min_band": 0}


def _set_switch(name: str, fn: str, v: int) -> int:
    """Set a tuning switch in libconv2d_tune.so; the entry points of this module call the tuning
    library while any switch is non-zero, and the product library again once all are back to 0."""
    L = load_tuning()
    old = getattr(L, fn)(int(v))
    _switches[name] = int(v)
    use_tuning_library(any(_switches.values()))
    return old


def debug_set_variant(v: int) -> int:
    """Tuning library only (not in include/conv2d.h): force a single-channel kernel variant; 0 = default."""
    return _set_switch("variant", "c2d_debug_set_variant", v)


def debug_set_min_band(v: int) -> int:
    """Tuning library only: minimum band height of the automatic band choice; 0 = default."""
    return _set_switch("min_band", "c2d_debug_set_min_band", v)


def debug_set_multi_variant(v: int) -> int:
    """Tuning library only: force a multi-channel kernel variant; 0 = default."""
    return _set_switch("multi_variant", "c2d_debug_set_multi_variant", v)

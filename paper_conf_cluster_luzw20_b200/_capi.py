"""ctypes binding of libconv2d.so -- the C ABI of include/conv2d.h, same names, argument marshalling
only. Loading fails loudly if the library is missing (there is no CPU or PyTorch fallback)."""
from __future__ import annotations

import ctypes
import os

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "libconv2d.so")

# every symbol include/conv2d.h declares
EXPORTS = ("conv2d_single", "conv2d_multi", "conv2d_single_ex", "conv2d_multi_ex", "conv2d_single_halo",
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


class Conv2dError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"{msg} (code {code})")
        self.code = code


def load(path: str | None = None):
    """Load libconv2d.so (built in-tree by __graft_entry__.build()). Raises if it is missing."""
    global _lib
    if _lib is not None:
        return _lib
    p = path or os.environ.get("C2D_LIB") or LIB_PATH  # C2D_LIB: tuning builds (tools/) only
    if not os.path.exists(p):
        raise ImportError(f"{p} is missing: run `python -c 'import __graft_entry__ as g; g.build()'` "
                          "(there is no fallback implementation)")
    L = ctypes.CDLL(p)
    P, I = ctypes.c_void_p, ctypes.c_int
    L.conv2d_single.argtypes = [P, I, I, P, I, P, P]
    L.conv2d_single_ex.argtypes = [P, I, I, P, I, P, P, I]
    if path is None and "C2D_LIB" in os.environ and not hasattr(L, "conv2d_single_halo"):
        pass  # an older tuning build (A/B timing only)
    else:
        L.conv2d_single_halo.argtypes = [P, I, I, P, I, P, I, P, P]
    if hasattr(L, "conv2d_single_pad"):
        L.conv2d_single_pad.argtypes = [P, I, I, P, I, I, P, P]
    L.conv2d_single_direct.argtypes = [P, I, I, P, I, P, P]
    L.conv2d_multi.argtypes = [P, I, I, I, I, P, I, I, P, P]
    L.conv2d_multi_ex.argtypes = [P, I, I, I, I, P, I, I, P, P, I]
    L.conv2d_single_host.argtypes = [P, I, I, P, I, P, P, I]
    L.conv2d_multi_tc.argtypes = [P, I, I, I, I, P, I, I, P, P]
    L.conv2d_release_scratch.argtypes = []
    for f in ("conv2d_single", "conv2d_single_ex", "conv2d_single_halo", "conv2d_single_pad", "conv2d_single_direct", "conv2d_multi",
              "conv2d_multi_ex", "conv2d_single_host", "conv2d_multi_tc", "conv2d_release_scratch",
              "conv2d_version"):
        if hasattr(L, f):
            getattr(L, f).restype = I
    L.conv2d_strerror.argtypes = [I]
    L.conv2d_strerror.restype = ctypes.c_char_p
    _lib = L
    return L


def lib():
    """The loaded library (hot path: one global lookup instead of load()'s checks)."""
    return _lib if _lib is not None else load()


def strerror(code: int) -> str:
    return load().conv2d_strerror(int(code)).decode()


def check(code: int) -> None:
    if code != CONV2D_OK:
        raise Conv2dError(code, strerror(code))


# raw entry points (device pointers as ints, stream handle as int): same names as the C ABI
def conv2d_single(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0) -> int:
    return load().conv2d_single(in_ptr, H, W, filt_ptr, K, out_ptr, stream)


def conv2d_single_ex(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0, band_h=0) -> int:
    return load().conv2d_single_ex(in_ptr, H, W, filt_ptr, K, out_ptr, stream, band_h)


def conv2d_single_pad(in_ptr, H, W, filt_ptr, K, mode, out_ptr, stream=0) -> int:
    return load().conv2d_single_pad(in_ptr, H, W, filt_ptr, K, mode, out_ptr, stream)


def conv2d_single_halo(in_ptr, H, W, halo_ptr, halo_rows, filt_ptr, K, out_ptr, stream=0) -> int:
    return load().conv2d_single_halo(in_ptr, H, W, halo_ptr, halo_rows, filt_ptr, K, out_ptr, stream)


def conv2d_single_direct(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0) -> int:
    return load().conv2d_single_direct(in_ptr, H, W, filt_ptr, K, out_ptr, stream)


def conv2d_multi(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream=0) -> int:
    return load().conv2d_multi(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream)


def conv2d_multi_ex(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream=0, band_h=0) -> int:
    return load().conv2d_multi_ex(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream, band_h)


def conv2d_single_host(in_ptr, H, W, filt_ptr, K, out_ptr, stream=0, chunk_rows=0) -> int:
    return load().conv2d_single_host(in_ptr, H, W, filt_ptr, K, out_ptr, stream, chunk_rows)


def conv2d_multi_tc(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream=0) -> int:
    return load().conv2d_multi_tc(in_ptr, N, C, H, W, filt_ptr, F, K, out_ptr, stream)


def conv2d_release_scratch() -> int:
    return load().conv2d_release_scratch()


def conv2d_version() -> int:
    return load().conv2d_version()


def debug_set_variant(v: int) -> int:
    """Tuning hook (not in include/conv2d.h): force a single-channel kernel variant; 0 = default."""
    L = load()
    L.c2d_debug_set_variant.argtypes = [ctypes.c_int]
    L.c2d_debug_set_variant.restype = ctypes.c_int
    return L.c2d_debug_set_variant(int(v))


def debug_set_min_band(v: int) -> int:
    """Tuning hook (not in include/conv2d.h): minimum band height of the automatic band choice."""
    L = load()
    L.c2d_debug_set_min_band.argtypes = [ctypes.c_int]
    L.c2d_debug_set_min_band.restype = ctypes.c_int
    return L.c2d_debug_set_min_band(int(v))


def debug_set_multi_variant(v: int) -> int:
    """Tuning hook (not in include/conv2d.h): force a multi-channel kernel variant; 0 = default."""
    L = load()
    L.c2d_debug_set_multi_variant.argtypes = [ctypes.c_int]
    L.c2d_debug_set_multi_variant.restype = ctypes.c_int
    return L.c2d_debug_set_multi_variant(int(v))

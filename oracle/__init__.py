"""CPU oracle for direct, stride-1, valid-mode fp32 2D convolution -- TEST INFRASTRUCTURE ONLY.

Only tests/, __graft_entry__.smoke() and bench.py (cpu_baseline leg and --impl reference) may import
this package. The product path (paper_conf_cluster_luzw20_b200/) never imports it; the two share no
code. See conv2d_oracle.c for the definition and its citations, paper_algorithms.py for the
step-by-step replays of the paper's Algorithms 1 and 2.

Every oracle function is pinned by tests/test_oracle.py (closed forms, textbook routines, brute
force, golden fixtures from the paper's worked examples). Parity unpinned: nothing -- except the
paper's performance numbers, which are relative speedups on other hardware.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "conv2d_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lib = None

_P = ctypes.c_void_p
_I = ctypes.c_int64


def build(force: bool = False) -> str:
    """Compile conv2d_oracle.c into liboracle.so (plain C, OpenMP, no fast-math, no contraction)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.run(["gcc", "-O2", "-std=c11", "-fopenmp", "-ffp-contract=off", "-fno-fast-math",
                        "-fPIC", "-shared", "-o", tmp, _SRC, "-lm"], check=True)
        os.replace(tmp, _LIB)
    return _LIB


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB)
        L.oracle_num_threads.restype = ctypes.c_int
        L.oracle_conv2d_single_rows.argtypes = [_P, _I, _I, _P, _I, _I, _I, _P, _P, _P]
        L.oracle_conv2d_single.argtypes = [_P, _I, _I, _P, _I, _P, _P, _P]
        L.oracle_conv2d_single_rect.argtypes = [_P, _I, _I, _P, _I, _I, _P, _P, _P]
        L.oracle_conv2d_single_points.argtypes = [_P, _I, _I, _P, _I, _P, _P, _I, _P, _P]
        L.oracle_conv2d_multi_images.argtypes = [_P, _I, _I, _I, _I, _P, _I, _I, _I, _I, _P, _P, _P]
        L.oracle_conv2d_multi.argtypes = [_P, _I, _I, _I, _I, _P, _I, _I, _P, _P, _P]
        L.oracle_conv2d_multi_points.argtypes = [_P, _I, _I, _I, _I, _P, _I, _I, _P, _P, _P, _P, _I,
                                                 _P, _P]
        _lib = L
    return _lib


def num_threads() -> int:
    return int(lib().oracle_num_threads())


def _ptr(a):
    return None if a is None else a.ctypes.data_as(ctypes.c_void_p)


def _f32(a):
    return np.ascontiguousarray(a, dtype=np.float32)


def conv2d_single(image, filt, want_bound=True, want_f64=False, rows=None):
    """Plain-definition single-channel valid cross-correlation (conv2d_oracle.c).

    image: H x W fp32; filt: K x K fp32. Returns (out fp32 [Ho x Wo], bound f64 or None,
    out64 f64 or None). `rows=(y0, y1)` restricts the computation to output rows [y0, y1): the other
    rows of the returned arrays are left uninitialised (bench cpu_baseline sample).
    """
    image = _f32(image)
    filt = _f32(filt)
    H, W = image.shape
    K = filt.shape[0]
    assert filt.shape == (K, K) and H >= K and W >= K
    Ho, Wo = H - K + 1, W - K + 1
    out = np.empty((Ho, Wo), np.float32)
    bound = np.empty((Ho, Wo), np.float64) if want_bound else None
    out64 = np.empty((Ho, Wo), np.float64) if want_f64 else None
    y0, y1 = (0, Ho) if rows is None else rows
    lib().oracle_conv2d_single_rows(_ptr(image), H, W, _ptr(filt), K, y0, y1, _ptr(out), _ptr(bound),
                                    _ptr(out64))
    return out, bound, out64


def conv2d_single_rect(image, filt, want_bound=True, want_f64=False):
    """Plain-definition valid cross-correlation with a rectangular FH x FW filter (conv2d_oracle.c
    oracle_conv2d_single_rect). Returns (out fp32, bound f64 or None, out64 or None)."""
    image = _f32(image)
    filt = _f32(filt)
    H, W = image.shape
    FH, FW = filt.shape
    assert H >= FH and W >= FW
    Ho, Wo = H - FH + 1, W - FW + 1
    out = np.empty((Ho, Wo), np.float32)
    bound = np.empty((Ho, Wo), np.float64) if want_bound else None
    out64 = np.empty((Ho, Wo), np.float64) if want_f64 else None
    lib().oracle_conv2d_single_rect(_ptr(image), H, W, _ptr(filt), FH, FW, _ptr(out), _ptr(bound), _ptr(out64))
    return out, bound, out64


def conv2d_single_points(image, filt, ys, xs):
    """Outputs at points (ys[p], xs[p]) computed one by one. Returns (out fp32, bound f64)."""
    image = _f32(image)
    filt = _f32(filt)
    H, W = image.shape
    K = filt.shape[0]
    ys = np.ascontiguousarray(ys, dtype=np.int64)
    xs = np.ascontiguousarray(xs, dtype=np.int64)
    assert ys.shape == xs.shape
    assert (ys >= 0).all() and (ys < H - K + 1).all() and (xs >= 0).all() and (xs < W - K + 1).all()
    out = np.empty(ys.shape, np.float32)
    bound = np.empty(ys.shape, np.float64)
    lib().oracle_conv2d_single_points(_ptr(image), H, W, _ptr(filt), K, _ptr(ys), _ptr(xs), ys.size,
                                      _ptr(out), _ptr(bound))
    return out, bound


def conv2d_multi(inp, filt, want_bound=True, want_f64=False, images=None):
    """Plain-definition multi-channel valid cross-correlation.

    inp: N x C x H x W; filt: F x C x K x K. Returns (out [N x F x Ho x Wo] fp32, bound, out64).
    `images=(n0, n1)` restricts to images [n0, n1) (others uninitialised).
    """
    inp = _f32(inp)
    filt = _f32(filt)
    N, C, H, W = inp.shape
    F, C2, K, K2 = filt.shape
    assert C2 == C and K2 == K and H >= K and W >= K
    Ho, Wo = H - K + 1, W - K + 1
    out = np.empty((N, F, Ho, Wo), np.float32)
    bound = np.empty((N, F, Ho, Wo), np.float64) if want_bound else None
    out64 = np.empty((N, F, Ho, Wo), np.float64) if want_f64 else None
    n0, n1 = (0, N) if images is None else images
    lib().oracle_conv2d_multi_images(_ptr(inp), N, C, H, W, _ptr(filt), F, K, n0, n1, _ptr(out),
                                     _ptr(bound), _ptr(out64))
    return out, bound, out64


def conv2d_multi_points(inp, filt, ns, fs, ys, xs):
    inp = _f32(inp)
    filt = _f32(filt)
    N, C, H, W = inp.shape
    F, _, K, _ = filt.shape
    arrs = [np.ascontiguousarray(a, dtype=np.int64) for a in (ns, fs, ys, xs)]
    n = arrs[0].size
    out = np.empty(n, np.float32)
    bound = np.empty(n, np.float64)
    lib().oracle_conv2d_multi_points(_ptr(inp), N, C, H, W, _ptr(filt), F, K, *[_ptr(a) for a in arrs],
                                     n, _ptr(out), _ptr(bound))
    return out, bound


def extend_image(image, K, padding):
    """The image extended by K-1 rows and columns for 'same' output (reading R20):
    E[r][c] = image[r - pt][c - pl] with pt = pl = (K-1)//2 (bottom / right get K-1-(K-1)//2, the
    torch padding='same' placement); outside the image E is 0 ("same_zero") or the nearest edge
    element ("same_replicate"). Written as an index map, element by element."""
    image = _f32(image)
    H, W = image.shape
    pt = (K - 1) // 2
    rows = np.arange(H + K - 1) - pt
    cols = np.arange(W + K - 1) - pt
    if padding == "same_replicate":
        return image[np.clip(rows, 0, H - 1)][:, np.clip(cols, 0, W - 1)]
    assert padding == "same_zero"
    E = np.zeros((H + K - 1, W + K - 1), np.float32)
    ri = (rows >= 0) & (rows < H)
    ci = (cols >= 0) & (cols < W)
    E[np.ix_(ri, ci)] = image
    return E


def conv2d_single_pad(image, filt, padding="valid", flip=False):
    """Boundary / semantic variants (include/conv2d.h conv2d_single_pad):

        out[y][x] = fl32( sum_i sum_j E[y+i][x+j] * g[i][j] )

    with E the image itself ("valid") or extend_image(...) ("same_zero", "same_replicate"), and
    g = filt (cross-correlation, the paper's orientation, R1) or g[i][j] = filt[K-1-i][K-1-j] (true
    convolution, flip=True: the NPP / ArrayFire orientation). The sum is the plain
    definition of conv2d_single above. Returns (out, bound, None)."""
    filt = _f32(filt)
    K = filt.shape[0]
    g = filt[::-1, ::-1] if flip else filt
    E = _f32(image) if padding == "valid" else extend_image(image, K, padding)
    return conv2d_single(E, g)


def within_tolerance(gpu, ref, bound, rel=1e-5):
    """The BASELINE.json north_star acceptance test |gpu - ref| <= rel * sum|x||w|, elementwise.

    Returns a boolean array. Equal values (including equal infinities / both NaN) always pass.
    """
    gpu = np.asarray(gpu, dtype=np.float64)
    ref = np.asarray(ref, dtype=np.float64)
    bound = np.asarray(bound, dtype=np.float64)
    with np.errstate(invalid="ignore"):
        ok = np.abs(gpu - ref) <= rel * bound
    same = (gpu == ref) | (np.isnan(gpu) & np.isnan(ref))
    return ok | same

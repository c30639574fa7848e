"""Pins of the CPU oracle (oracle/conv2d_oracle.c) against things other than itself.

Closed forms (impulse, delta filter, K=1, constant input, box filter vs summed-area table), exactness
with integer data, textbook/library routines on tiny inputs (scipy.signal.correlate2d, float64
torch.nn.functional.conv2d), invariants (linearity, separability, channel decomposition, NaN
receptive field), and the sampled/row-range entry points against the full computation.
"""
import numpy as np
import pytest
import scipy.signal
import torch

import oracle
from gen import synth

RNG = np.random.default_rng(20200914)


def _img(H, W, dist="sym", seed=1):
    return synth.fill_np(seed, synth.TAG_INPUT, (H, W), dist)


def _flt(K, dist="rand", seed=2):
    return synth.make_filter(seed, K, dist)[0, 0]


# ---------------------------------------------------------------- closed forms (bitwise)
@pytest.mark.parametrize("K", [1, 2, 3, 5, 8, 15])
def test_impulse_input_gives_filter(K):
    """in = e_(r0,c0) => out[y][x] = f[r0-y][c0-x] inside the range, else 0 (orientation: no flip)."""
    H, W = K + 9, K + 7
    f = _flt(K, "rand", seed=K)
    for (r0, c0) in [(0, 0), (K - 1, K - 1), (H // 2, W // 3), (H - 1, W - 1)]:
        img = np.zeros((H, W), np.float32)
        img[r0, c0] = 1.0
        out, _, _ = oracle.conv2d_single(img, f)
        exp = np.zeros_like(out)
        for y in range(out.shape[0]):
            for x in range(out.shape[1]):
                i, j = r0 - y, c0 - x
                if 0 <= i < K and 0 <= j < K:
                    exp[y, x] = f[i, j]
        assert np.array_equal(out.view(np.uint32), exp.view(np.uint32))


@pytest.mark.parametrize("K", [1, 3, 4, 7, 15])
def test_delta_filter_is_shift(K):
    """f = e_(i0,j0) => out[y][x] = in[y+i0][x+j0] (BASELINE.json north_star closed form)."""
    H, W = 2 * K + 5, 3 * K + 2
    img = _img(H, W, "img", seed=K)
    Ho, Wo = H - K + 1, W - K + 1
    for (i0, j0) in {(0, 0), (K - 1, 0), (0, K - 1), (K // 2, K // 2), (K - 1, K - 1)}:
        f = np.zeros((K, K), np.float32)
        f[i0, j0] = 1.0
        out, _, _ = oracle.conv2d_single(img, f)
        assert np.array_equal(out, img[i0:i0 + Ho, j0:j0 + Wo])


def test_k1_is_correctly_rounded_scale():
    img = _img(33, 41, "sym")
    for w in (np.float32(0.3), np.float32(-1.7e-3), np.float32(3.0)):
        out, _, _ = oracle.conv2d_single(img, np.array([[w]], np.float32))
        assert np.array_equal(out, img * w)  # IEEE fp32 product = one rounding of the exact product


@pytest.mark.parametrize("K", [2, 3, 5, 9, 15])
def test_constant_input(K):
    """in == c => out == c * sum(w) exactly for dyadic c and small-integer w."""
    c = np.float32(0.75)
    f = synth.make_filter(K, K, "int")[0, 0]
    img = np.full((K + 6, K + 11), c, np.float32)
    out, _, _ = oracle.conv2d_single(img, f)
    assert (out == np.float32(float(c) * float(f.astype(np.float64).sum()))).all()


@pytest.mark.parametrize("K", [1, 3, 6, 11, 15])
def test_box_filter_matches_summed_area_table(K):
    """Box filter == prefix-sum result S[y+K][x+K] - S[y][x+K] - S[y+K][x] + S[y][x] (int64)."""
    H, W = K + 20, K + 17
    img = _img(H, W, "int", seed=K)
    S = np.zeros((H + 1, W + 1), np.int64)
    S[1:, 1:] = img.astype(np.int64).cumsum(0).cumsum(1)
    exp = S[K:, K:] - S[:-K, K:] - S[K:, :-K] + S[:-K, :-K]
    out, _, _ = oracle.conv2d_single(img, np.ones((K, K), np.float32))
    assert np.array_equal(out, exp.astype(np.float32))


def test_integer_data_exact():
    """Integer data: every partial sum is an exactly representable integer -> exact result."""
    for K in (3, 7, 15):
        img = _img(K + 13, K + 9, "int", seed=K)
        f = synth.make_filter(K, K, "int")[0, 0]
        out, bound, out64 = oracle.conv2d_single(img, f, want_f64=True)
        ref = np.zeros(out.shape, np.int64)
        for y in range(out.shape[0]):
            for x in range(out.shape[1]):
                ref[y, x] = int((img[y:y + K, x:x + K].astype(np.int64) * f.astype(np.int64)).sum())
        assert np.array_equal(out64, ref.astype(np.float64))
        assert np.array_equal(out, ref.astype(np.float32))
        assert (bound >= np.abs(out64)).all()


# ---------------------------------------------------------------- textbook / library routines
def test_matches_scipy_correlate2d_bruteforce():
    """Tiny inputs, K = 1..15, H, W in [K, K+6]: out64 == scipy.signal.correlate2d(valid)."""
    for K in range(1, 16):
        for trial in range(3):
            H = K + int(RNG.integers(0, 7))
            W = K + int(RNG.integers(0, 7))
            img = RNG.standard_normal((H, W)).astype(np.float32)
            f = RNG.standard_normal((K, K)).astype(np.float32)
            out, bound, out64 = oracle.conv2d_single(img, f, want_f64=True)
            ref = scipy.signal.correlate2d(img.astype(np.float64), f.astype(np.float64), mode="valid")
            assert ref.shape == out.shape
            assert (np.abs(out64 - ref) <= 1e-12 * bound).all()
            assert np.array_equal(out, out64.astype(np.float32))  # exactly one rounding
            ab = scipy.signal.correlate2d(np.abs(img.astype(np.float64)), np.abs(f.astype(np.float64)),
                                          mode="valid")
            assert np.allclose(bound, ab, rtol=1e-12, atol=0)


def test_multi_matches_torch_conv2d_float64():
    """Multi-channel oracle == float64 torch.nn.functional.conv2d (OIHW, cross-correlation)."""
    for (N, C, F, K, H, W) in [(1, 1, 1, 3, 7, 9), (2, 3, 4, 5, 11, 8), (2, 4, 3, 7, 9, 13),
                               (1, 2, 2, 1, 4, 4), (3, 3, 2, 15, 16, 18), (1, 4, 5, 4, 10, 6)]:
        inp = RNG.standard_normal((N, C, H, W)).astype(np.float32)
        w = RNG.standard_normal((F, C, K, K)).astype(np.float32)
        out, bound, out64 = oracle.conv2d_multi(inp, w, want_f64=True)
        ref = torch.nn.functional.conv2d(torch.from_numpy(inp).double(), torch.from_numpy(w).double())
        assert (np.abs(out64 - ref.numpy()) <= 1e-12 * bound).all()
        assert np.array_equal(out, out64.astype(np.float32))


# ---------------------------------------------------------------- invariants
def test_linearity():
    K = 5
    x = _img(30, 31, "sym", 1)
    y = _img(30, 31, "sym", 2)
    f = _flt(K)
    a, b = 1.0, -1.0  # sym values are k/2^23 with |k| <= 2^23: x - y is exact in fp32
    z = (a * x.astype(np.float64) + b * y.astype(np.float64)).astype(np.float32)
    assert np.array_equal(z.astype(np.float64), a * x.astype(np.float64) + b * y.astype(np.float64))
    _, bz, oz = oracle.conv2d_single(z, f, want_f64=True)
    _, _, ox = oracle.conv2d_single(x, f, want_f64=True)
    _, _, oy = oracle.conv2d_single(y, f, want_f64=True)
    assert (np.abs(oz - (a * ox + b * oy)) <= 1e-12 * (bz + 1)).all()
    _, _, o4 = oracle.conv2d_single(x * np.float32(4.0), f, want_f64=True)  # exact power-of-2 scale
    assert np.array_equal(o4, 4.0 * ox)


def test_separable_filter():
    """f = u v^T: conv == column pass by u of the row pass by v."""
    K = 7
    u = RNG.standard_normal(K).astype(np.float32)
    v = RNG.standard_normal(K).astype(np.float32)
    f = np.outer(u.astype(np.float64), v.astype(np.float64))
    f32 = f.astype(np.float32)
    img = _img(40, 37, "sym")
    _, bound, o64 = oracle.conv2d_single(img, f32, want_f64=True)
    rows = np.stack([np.correlate(r.astype(np.float64), v.astype(np.float64), "valid") for r in img])
    sep = np.stack([np.correlate(c, u.astype(np.float64), "valid") for c in rows.T]).T
    # f32 = f rounded: allow the filter rounding (2^-24 relative per tap) in the comparison
    assert (np.abs(o64 - sep) <= 1e-6 * bound).all()


def test_multi_is_sum_over_channels_and_reduces_to_single():
    N, C, F, K, H, W = 2, 3, 2, 4, 12, 15
    inp = synth.fill_np(4, 1, (N, C, H, W), "sym")
    w = synth.make_filter(4, K, "rand", F=F, C=C)
    out, bound, out64 = oracle.conv2d_multi(inp, w, want_f64=True)
    for n in range(N):
        for f in range(F):
            s = sum(oracle.conv2d_single(inp[n, c], w[f, c], want_f64=True)[2] for c in range(C))
            assert (np.abs(out64[n, f] - s) <= 1e-12 * bound[n, f]).all()
    o1, _, _ = oracle.conv2d_multi(inp[:1, :1], w[:1, :1])
    s1, _, _ = oracle.conv2d_single(inp[0, 0], w[0, 0])
    assert np.array_equal(o1[0, 0], s1)


def test_nan_receptive_field():
    """A NaN at (r, c) poisons exactly outputs y in [r-K+1, r], x in [c-K+1, c]."""
    K, H, W = 5, 20, 23
    img = _img(H, W, "img")
    r, c = 9, 11
    img[r, c] = np.nan
    out, _, _ = oracle.conv2d_single(img, _flt(K))
    mask = np.zeros(out.shape, bool)
    mask[max(0, r - K + 1):r + 1, max(0, c - K + 1):c + 1] = True
    assert np.array_equal(np.isnan(out), mask)


# ---------------------------------------------------------------- entry points agree
def test_points_and_rows_match_full():
    K = 6
    img = _img(50, 61, "img")
    f = _flt(K)
    out, bound, _ = oracle.conv2d_single(img, f)
    ys = RNG.integers(0, out.shape[0], 200)
    xs = RNG.integers(0, out.shape[1], 200)
    po, pb = oracle.conv2d_single_points(img, f, ys, xs)
    assert np.array_equal(po, out[ys, xs]) and np.array_equal(pb, bound[ys, xs])
    ro, _, _ = oracle.conv2d_single(img, f, rows=(7, 19))
    assert np.array_equal(ro[7:19], out[7:19])

    inp = synth.fill_np(9, 1, (3, 2, 14, 17), "sym")
    w = synth.make_filter(9, 3, "he", F=4, C=2)
    mo, mb, _ = oracle.conv2d_multi(inp, w)
    n, fi, y, x = (RNG.integers(0, s, 100) for s in mo.shape)
    qo, qb = oracle.conv2d_multi_points(inp, w, n, fi, y, x)
    assert np.array_equal(qo, mo[n, fi, y, x]) and np.array_equal(qb, mb[n, fi, y, x])
    io, _, _ = oracle.conv2d_multi(inp, w, images=(1, 3))
    assert np.array_equal(io[1:3], mo[1:3])


def test_within_tolerance_helper():
    ref = np.array([1.0, 2.0, np.nan, 0.0])
    bound = np.array([1.0, 1.0, 1.0, 0.0])
    assert oracle.within_tolerance(ref + [1e-6, 0, 0, 0], ref, bound).tolist() == [True, True, True, True]
    assert not oracle.within_tolerance(ref + [2e-5, 0, 0, 0], ref, bound)[0]
    assert not oracle.within_tolerance(ref + [0, 0, 0, 1e-30], ref, bound)[3]



# ---------------------------------------------------------------------------------------------
# N4 boundary / semantic variants (oracle.conv2d_single_pad)
# ---------------------------------------------------------------------------------------------
@pytest.mark.parametrize("K", [1, 2, 3, 4, 5, 8, 15])
def test_same_zero_matches_torch_padding_same(K):
    """'same' zero padding (both odd and even K) == torch.nn.functional.conv2d(padding='same') in f64."""
    import torch

    rng = np.random.default_rng(K)
    for (H, W) in [(K + 5, K + 9), (3, 4), (1, 1), (17, 2)]:
        x = rng.standard_normal((H, W)).astype(np.float32)
        f = rng.standard_normal((K, K)).astype(np.float32)
        y, bound, _ = oracle.conv2d_single_pad(x, f, "same_zero")
        ref = torch.nn.functional.conv2d(torch.from_numpy(x).double()[None, None], torch.from_numpy(f).double()[None, None],
                                         padding="same")[0, 0].numpy()
        assert y.shape == (H, W)
        assert np.allclose(y, ref, rtol=0, atol=1e-6 * (1 + np.abs(ref).max()))


@pytest.mark.parametrize("K", [2, 3, 6, 7])
def test_same_replicate_matches_torch_replicate_pad(K):
    import torch

    rng = np.random.default_rng(K + 100)
    x = rng.standard_normal((K + 7, K + 3)).astype(np.float32)
    f = rng.standard_normal((K, K)).astype(np.float32)
    y, _, _ = oracle.conv2d_single_pad(x, f, "same_replicate")
    pt = (K - 1) // 2
    xp = torch.nn.functional.pad(torch.from_numpy(x).double()[None, None], (pt, K - 1 - pt, pt, K - 1 - pt),
                                 mode="replicate")
    ref = torch.nn.functional.conv2d(xp, torch.from_numpy(f).double()[None, None])[0, 0].numpy()
    assert np.allclose(y, ref, rtol=0, atol=1e-6 * (1 + np.abs(ref).max()))


@pytest.mark.parametrize("K", [1, 3, 4, 9])
def test_flip_matches_scipy_convolve2d(K):
    """True convolution == scipy.signal.convolve2d (valid), the textbook flipped-kernel definition."""
    from scipy.signal import convolve2d

    rng = np.random.default_rng(K + 7)
    x = rng.standard_normal((K + 6, K + 11)).astype(np.float32)
    f = rng.standard_normal((K, K)).astype(np.float32)
    y, _, _ = oracle.conv2d_single_pad(x, f, "valid", flip=True)
    ref = convolve2d(x.astype(np.float64), f.astype(np.float64), mode="valid")
    assert np.allclose(y, ref, rtol=0, atol=1e-6 * (1 + np.abs(ref).max()))


@pytest.mark.parametrize("K", [1, 3, 5, 15])
def test_same_zero_centered_delta_is_identity(K):
    """odd K, 'same' zero padding, delta at the centre: every output equals its input (bitwise)."""
    x = synth.fill_np(5, synth.TAG_INPUT, (K + 4, 2 * K + 3), "sym")
    f = np.zeros((K, K), np.float32)
    f[K // 2, K // 2] = 1.0
    y, _, _ = oracle.conv2d_single_pad(x, f, "same_zero")
    assert np.array_equal(y, x)


@pytest.mark.parametrize("K", [2, 5, 8])
def test_same_zero_box_filter_counts_window_cells(K):
    """ones image, box filter, zero padding: out[y][x] = (#rows of the window inside the image) *
    (#columns inside) -- a closed form of the padding placement (top/left (K-1)//2)."""
    H, W = K + 3, 2 * K + 1
    y, _, _ = oracle.conv2d_single_pad(np.ones((H, W), np.float32), np.ones((K, K), np.float32), "same_zero")
    pt = (K - 1) // 2

    def inside(n, L):
        return np.array([sum(1 for i in range(K) if 0 <= v + i - pt < L) for v in range(n)], np.float64)

    assert np.array_equal(y, np.outer(inside(H, H), inside(W, W)).astype(np.float32))


@pytest.mark.parametrize("K", [3, 4, 7])
def test_same_replicate_constant_image(K):
    """replicate padding of a constant image is the constant everywhere: out = c * sum(w), exactly
    (small integers)."""
    f = np.arange(K * K, dtype=np.float32).reshape(K, K) - 5
    y, _, _ = oracle.conv2d_single_pad(np.full((K + 2, K + 5), 3.0, np.float32), f, "same_replicate")
    assert np.array_equal(y, np.full(y.shape, 3.0 * f.sum(), np.float32))


@pytest.mark.parametrize("K", [2, 3, 6])
def test_flip_impulse_gives_filter_upright(K):
    """true convolution of an impulse at (r0, c0) is the filter in its own orientation at
    [r0-K+1, r0] x [c0-K+1, c0] (cross-correlation gives it rotated: test_impulse_input_gives_filter)."""
    H, W = 3 * K, 3 * K + 1
    r0, c0 = K + 1, K + 2
    x = np.zeros((H, W), np.float32)
    x[r0, c0] = 1.0
    f = synth.make_filter(3, K, "rand")[0, 0]
    y, _, _ = oracle.conv2d_single_pad(x, f, "valid", flip=True)
    exp = np.zeros_like(y)
    exp[r0 - K + 1:r0 + 1, c0 - K + 1:c0 + 1] = f
    assert np.array_equal(y, exp)


# --------------------------------------------------------------------------------------------
# Rectangular FH x FW filters (Table I's "FH x FW" columns)
# --------------------------------------------------------------------------------------------
RECT_SHAPES = [(1, 5), (5, 1), (3, 7), (7, 3), (2, 15), (15, 2), (4, 9), (13, 6)]


def test_rect_matches_scipy_correlate2d_bruteforce():
    """Textbook routine: scipy.signal.correlate2d(mode='valid') in float64 on tiny shapes."""
    import scipy.signal

    rng = np.random.default_rng(7)
    for FH, FW in RECT_SHAPES:
        for dh, dw in [(0, 0), (1, 3), (6, 2)]:
            x = rng.standard_normal((FH + dh, FW + dw)).astype(np.float32)
            f = rng.standard_normal((FH, FW)).astype(np.float32)
            y, bound, y64 = oracle.conv2d_single_rect(x, f, want_f64=True)
            ref = scipy.signal.correlate2d(x.astype(np.float64), f.astype(np.float64), mode="valid")
            assert y.shape == ref.shape == (dh + 1, dw + 1)
            assert np.all(np.abs(y64 - ref) <= 1e-12 * bound)
            assert np.array_equal(y, ref.astype(np.float32))


def test_rect_delta_filter_is_shift():
    """Closed form: a delta at (i0, j0) of an FH x FW filter shifts the image by (i0, j0)."""
    x = synth.fill_np(3, synth.TAG_INPUT, (30, 41), "sym")
    for FH, FW in RECT_SHAPES:
        for i0, j0 in [(0, 0), (FH - 1, FW - 1), (FH // 2, FW - 1)]:
            f = np.zeros((FH, FW), np.float32)
            f[i0, j0] = 1.0
            y, _, _ = oracle.conv2d_single_rect(x, f)
            assert np.array_equal(y, x[i0:i0 + 30 - FH + 1, j0:j0 + 41 - FW + 1])


def test_rect_box_filter_matches_summed_area_table():
    """Closed form: an all-ones FH x FW filter on integer data sums the FH x FW window (prefix sums)."""
    x = synth.fill_np(5, synth.TAG_INPUT, (40, 50), "int").astype(np.int64)
    S = np.zeros((41, 51), np.int64)
    S[1:, 1:] = x.cumsum(0).cumsum(1)
    for FH, FW in RECT_SHAPES:
        y, _, _ = oracle.conv2d_single_rect(x.astype(np.float32), np.ones((FH, FW), np.float32))
        ref = S[FH:, FW:] - S[:-FH, FW:] - S[FH:, :-FW] + S[:-FH, :-FW]
        assert np.array_equal(y, ref.astype(np.float32))


def test_rect_square_reduces_to_single_and_transpose_swaps_shape():
    """Invariants: FH == FW is the square definition; correlating the transposed image with the
    transposed filter gives the transposed output (catches an FH/FW or i/j swap)."""
    x = synth.fill_np(9, synth.TAG_INPUT, (33, 47), "img")
    for K in (1, 4, 9):
        f = synth.make_filter(9, K, "rand")[0, 0]
        assert np.array_equal(oracle.conv2d_single_rect(x, f)[0], oracle.conv2d_single(x, f)[0])
    rng = np.random.default_rng(3)
    for FH, FW in RECT_SHAPES:
        f = rng.standard_normal((FH, FW)).astype(np.float32)
        y, _, _ = oracle.conv2d_single_rect(x, f)
        yt, _, _ = oracle.conv2d_single_rect(np.ascontiguousarray(x.T), np.ascontiguousarray(f.T))
        assert yt.shape == y.T.shape
        assert np.allclose(yt, y.T, rtol=1e-6, atol=1e-6)


def test_rect_separable_filter():
    """Closed form: f = u v^T (FH x 1 times 1 x FW) is a column correlation by u after a row
    correlation by v."""
    x = synth.fill_np(11, synth.TAG_INPUT, (25, 31), "sym")
    rng = np.random.default_rng(11)
    for FH, FW in RECT_SHAPES:
        u = rng.integers(-3, 4, (FH, 1)).astype(np.float32)
        v = rng.integers(-3, 4, (1, FW)).astype(np.float32)
        xi = np.round(x * 8).astype(np.float32)  # integers: every order exact
        rows, _, _ = oracle.conv2d_single_rect(xi, v)
        both, _, _ = oracle.conv2d_single_rect(rows, u)
        direct, _, _ = oracle.conv2d_single_rect(xi, u @ v)
        assert np.array_equal(both, direct)

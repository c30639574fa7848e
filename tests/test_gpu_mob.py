"""GPU tests of the filter-blocked multi-channel kernel (conv2d_mob.cuh, the conv2d_multi default):
every output against the CPU oracle on shapes that hit every path (segment widths 4-32 lanes, FB = 8 and
FB = 4, warp-steps spanning rows and images, idle segments in the last step, ragged right edges, the
misaligned-input instantiation, 16-/8-/4-byte output alignment, F not a multiple of the F-block),
integer data exact, and bitwise equality with the round-2 ring kernel (tuning variant 8) and across
every tuning shape of the kernel itself (variants 100-112) and every explicit tiling."""
import pytest
import torch

import paper_conf_cluster_luzw20_b200 as pkg
from gen import synth
from tests.gpu_helpers import check_full_multi, dev_image

pytestmark = pytest.mark.gpu
DEV = "cuda"
MOB_VARIANTS = [100, 101, 102, 103, 104, 105, 106, 107, 108, 109, 112]


def _w(F, C, K, dist="he", seed=5):
    return torch.from_numpy(synth.make_filter(seed, K, dist, F=F, C=C)).to(DEV)


# (N, C, F, H - K, W - K): narrow (4-lane segments), 54-wide (8), 100-wide, 218-wide, > 256-wide
SHAPES = [(3, 3, 13, 9, 21), (2, 5, 8, 20, 53), (1, 2, 17, 7, 99), (2, 3, 9, 6, 217), (1, 1, 20, 5, 300)]


@pytest.mark.parametrize("K", [1, 2, 3, 4, 5, 6, 7, 8, 9, 11, 15])
def test_default_vs_oracle(cuda_device, K):
    for (N, C, F, dh, dw) in SHAPES:
        x = dev_image((N, C, K + dh, K + dw), "sym", seed=K + C)
        w = _w(F, C, K, seed=K + F)
        check_full_multi(x, w, pkg.conv2d_multi(x, w))


@pytest.mark.parametrize("K", [1, 3, 5, 7, 9, 15])
def test_integer_exact_and_ring_kernel_bits(cuda_device, K):
    """Integer data: exact sums. Real data: the same bits as the round-2 ring kernel (variant 8), whose
    per-output order is the same (filter row, channel, filter column) fmaf chain."""
    from paper_conf_cluster_luzw20_b200 import _capi

    xi = dev_image((3, 3, K + 11, K + 70), "int", seed=K)
    wi = _w(10, 3, K, "int", seed=K)
    check_full_multi(xi, wi, pkg.conv2d_multi(xi, wi), exact=True)
    x = dev_image((3, 4, K + 13, K + 90), "img", seed=K + 1)
    w = _w(11, 4, K, seed=K + 1)
    y = pkg.conv2d_multi(x, w)
    try:
        _capi.debug_set_multi_variant(8)
        y8 = pkg.conv2d_multi(x, w)
    finally:
        _capi.debug_set_multi_variant(0)
    assert torch.equal(y, y8)


@pytest.mark.parametrize("K", [3, 5, 7])
def test_every_variant_and_tiling_bitwise(cuda_device, K):
    from paper_conf_cluster_luzw20_b200 import _capi

    for (N, C, F, dh, dw) in [(5, 3, 19, 12, 45), (2, 2, 8, 30, 150)]:
        x = dev_image((N, C, K + dh, K + dw), "img", seed=K + N)
        w = _w(F, C, K, seed=K + F)
        y = pkg.conv2d_multi(x, w)
        check_full_multi(x, w, y)
        for L in (1, 2, 7, 1000):  # explicit warp-steps per warp
            assert torch.equal(pkg.conv2d_multi(x, w, band_h=L), y), (K, L)
        try:
            for v in MOB_VARIANTS:
                _capi.debug_set_multi_variant(v)
                assert torch.equal(pkg.conv2d_multi(x, w), y), (K, v)
        finally:
            _capi.debug_set_multi_variant(0)


@pytest.mark.parametrize("K", [3, 7])
def test_alignment_paths(cuda_device, K):
    """Misaligned input rows (W % 4 != 0 and an offset base: the guarded scalar-load instantiation);
    output row pitch Wo % 4 in {0, 2, odd} and an offset output pointer (vector / 8-byte / scalar
    stores)."""
    for W in (K + 63, K + 61, K + 62, K + 64):  # Wo = 64 (16 B rows), 62 (8 B), 63 (odd), 65
        base = dev_image((2 * 3 * (K + 9) * W + 1,), "sym", seed=W)
        for off in (0, 1):
            x = base[off:off + 2 * 3 * (K + 9) * W].view(2, 3, K + 9, W)
            w = _w(6, 3, K, seed=W)
            y = pkg.conv2d_multi(x, w)
            check_full_multi(x, w, y)
            Ho, Wo = 9 + 1, W - K + 1
            buf = torch.empty(2 * 6 * Ho * Wo + 3, device=DEV)
            for oo in (1, 2):
                out = buf[oo:oo + 2 * 6 * Ho * Wo].view(2, 6, Ho, Wo)
                assert torch.equal(pkg.conv2d_multi(x, w, out=out), y), (K, W, off, oo)


def test_small_grid_takes_fb4(cuda_device):
    """A layer whose FB = 8 grid fills less than 3/4 of a wave (Table I CONV7 shape at N = 16) runs the
    FB = 4 form: same bits as FB = 8 (variant 100), oracle parity."""
    from paper_conf_cluster_luzw20_b200 import _capi

    x = dev_image((16, 3, 28, 28), "img", seed=7)
    w = _w(16, 3, 5, seed=7)
    y = pkg.conv2d_multi(x, w)
    check_full_multi(x, w, y)
    try:
        _capi.debug_set_multi_variant(100)
        y8 = pkg.conv2d_multi(x, w)
    finally:
        _capi.debug_set_multi_variant(0)
    assert torch.equal(y, y8)


def test_cuda_graph_capture_and_concurrent_streams(cuda_device):
    """conv2d_multi captured into a CUDA graph replays correctly and picks up new inputs and filters at
    replay; calls with different filters on three streams give the one-stream bits (the F-block is
    staged per CTA from the caller's filter tensor: no library-global state between calls)."""
    x = dev_image((6, 3, 60, 90), "img", seed=3)
    w = _w(20, 3, 5, seed=3)
    y = torch.empty((6, 20, 56, 86), device=DEV)
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        pkg.conv2d_multi(x, w, out=y)  # warm-up outside capture (occupancy and smem attributes)
    torch.cuda.current_stream().wait_stream(s)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        pkg.conv2d_multi(x, w, out=y)
    g.replay()
    torch.cuda.synchronize()
    check_full_multi(x, w, y)
    x.copy_(dev_image((6, 3, 60, 90), "sym", seed=4))
    w.copy_(_w(20, 3, 5, seed=4))
    g.replay()
    torch.cuda.synchronize()
    check_full_multi(x, w, y)

    ws = [_w(12, 3, 7, seed=10 + i) for i in range(6)]
    xs = dev_image((4, 3, 40, 230), "img", seed=11)
    outs = [torch.empty((4, 12, 34, 224), device=DEV) for _ in ws]
    streams = [torch.cuda.Stream() for _ in range(3)]
    for st in streams:
        st.wait_stream(torch.cuda.current_stream())
    for i, wi in enumerate(ws):
        st = streams[i % 3]
        with torch.cuda.stream(st):
            pkg.conv2d_multi(xs, wi, out=outs[i], stream=st)
    torch.cuda.synchronize()
    for wi, yi in zip(ws, outs):
        assert torch.equal(yi, pkg.conv2d_multi(xs, wi))


@pytest.mark.parametrize("C,K", [(40, 15), (200, 15), (300, 9)])
def test_large_c_fallback(cuda_device, C, K):
    """F-blocks beyond shared memory: C*K*K*8*4 B (FB = 8) or *4 (FB = 4) past the opt-in limit hand over
    to FB = 4 or to the round-1 kernel with one filter per warp (C*K*ceil(K/4)*16 B); every output
    against the oracle either way."""
    x = dev_image((1, C, K + 3, K + 40), "sym", seed=C)
    w = _w(5, C, K, seed=C)
    y = pkg.conv2d_multi(x, w)
    check_full_multi(x, w, y)

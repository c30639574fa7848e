"""GPU parity of conv2d_single (C ABI via the binding) against the CPU oracle.

Small shapes are compared element by element (all K in 1..15, ragged widths, every W % 4, Wo < 32,
H == K, W == K, misaligned pointers); the BASELINE.json configs at full size are compared element by
element too (every output of the 28 sweep points; configs[4]: every output around the 8-way row-band
seams and of two whole bands), in the launch configuration bench.py times.
"""
import numpy as np
import pytest
import torch

import paper_conf_cluster_luzw20_b200 as pkg
from gen import synth
from paper_conf_cluster_luzw20_b200 import _capi
from tests.gpu_helpers import check_full_single, check_full_single_host, dev_image

pytestmark = pytest.mark.gpu
DEV = "cuda"


def _filt(K, dist="rand", seed=3):
    return torch.from_numpy(synth.make_filter(seed, K, dist)[0, 0]).to(DEV)


def test_config0_256_k3(cuda_device):
    """BASELINE.json configs[0]: 256x256, 3x3, valid, stride 1 -- every output."""
    x = dev_image((256, 256), "img")
    for dist in ("rand", "gauss", "box"):
        f = _filt(3, dist)
        check_full_single(x, f, pkg.conv2d_single(x, f))


SMALL_SHAPES = [(0, 0), (1, 3), (9, 4), (37, 300), (70, 517), (33, 1023), (20, 1030), (150, 256)]


@pytest.mark.parametrize("K", list(range(1, 16)))
def test_all_k_small_shapes(cuda_device, K):
    rng = np.random.default_rng(K)
    for (dh, dw) in SMALL_SHAPES:
        H, W = K + dh, K + dw
        x = dev_image((H, W), "sym", seed=K * 1000 + dh)
        f = _filt(K, "rand", seed=K)
        check_full_single(x, f, pkg.conv2d_single(x, f))
    # one random non-trivial band height on a taller image: several bands and a ragged last band
    x = dev_image((K + 75, 389), "img", seed=K)
    f = _filt(K, "gauss")
    check_full_single(x, f, pkg.conv2d_single(x, f, band_h=int(rng.integers(1, 20))))


@pytest.mark.parametrize("K", [1, 2, 3, 4, 5, 7, 9, 11, 13, 15])
def test_integer_data_bitwise(cuda_device, K):
    """Integer data: every fp32 partial sum is exact, so the GPU must equal the oracle bit for bit."""
    for (H, W) in [(K + 40, 517), (K + 3, 1024), (2 * K + 1, 131)]:
        x = dev_image((H, W), "int", seed=H + K)
        f = _filt(K, "int", seed=K)
        check_full_single(x, f, pkg.conv2d_single(x, f), exact=True)


@pytest.mark.parametrize("K", [3, 5, 8, 15])
def test_misaligned_pointers(cuda_device, K):
    """in / out offset by 1..3 floats from 16-byte alignment take the scalar / shifted-store paths."""
    H, W = K + 50, 600
    for off_in in (0, 1, 2, 3):
        for off_out in (0, 1, 3):
            xb = dev_image((H * W + 4,), "img", seed=off_in)
            x = xb[off_in:off_in + H * W].view(H, W)
            ob = torch.empty((H - K + 1) * (W - K + 1) + 4, device=DEV)
            y = ob[off_out:off_out + (H - K + 1) * (W - K + 1)].view(H - K + 1, W - K + 1)
            f = _filt(K)
            pkg.conv2d_single(x, f, out=y)
            check_full_single(x, f, y)


@pytest.mark.parametrize("K", [1, 3, 6, 15])
def test_band_height_does_not_change_bits(cuda_device, K):
    """Every output's summation order is independent of its band (and so of any row-band shard)."""
    x = dev_image((K + 300, 700), "img", seed=K)
    f = _filt(K)
    ref = pkg.conv2d_single(x, f)
    for bh in (1, 2, 5, 17, 64, 10 ** 6):
        assert torch.equal(pkg.conv2d_single(x, f, band_h=bh), ref)
    # a row sub-range computed on its own (what a row-band shard does) equals the matching rows
    r0, r1 = 37, 201
    sub = pkg.conv2d_single(x[r0:r1 + K - 1].contiguous(), f)
    assert torch.equal(sub, ref[r0:r1])


def test_nan_receptive_field(cuda_device):
    K, H, W = 5, 80, 300
    x = dev_image((H, W), "img")
    r, c = 41, 133
    x[r, c] = float("nan")
    y = pkg.conv2d_single(x, _filt(K)).cpu().numpy()
    mask = np.zeros(y.shape, bool)
    mask[r - K + 1:r + 1, c - K + 1:c + 1] = True
    assert np.array_equal(np.isnan(y), mask)


def test_closed_forms_on_gpu(cuda_device):
    x = dev_image((200, 333), "img")
    for K in (3, 7, 15):
        d = torch.zeros((K, K), device=DEV)
        d[K // 2, K - 1] = 1.0
        y = pkg.conv2d_single(x, d)
        assert torch.equal(y, x[K // 2:K // 2 + 200 - K + 1, K - 1:K - 1 + 333 - K + 1])
    c = torch.full((64, 300), 0.75, device=DEV)
    f = _filt(9, "int")
    assert (pkg.conv2d_single(c, f) == 0.75 * float(f.double().sum())).all()


def test_direct_baseline_kernel(cuda_device):
    for K in (3, 5, 15):
        x = dev_image((K + 60, 257), "img", seed=K)
        f = _filt(K)
        check_full_single(x, f, pkg.conv2d_single_direct(x, f))


def test_error_codes_on_device(cuda_device):
    x = torch.zeros((10, 10), device=DEV)
    f = torch.zeros((3, 3), device=DEV)
    y = torch.zeros((8, 8), device=DEV)
    assert _capi.conv2d_single(x.data_ptr(), 10, 10, f.data_ptr(), 16, y.data_ptr()) == _capi.CONV2D_EK
    assert _capi.conv2d_single(x.data_ptr(), 10, 10, f.data_ptr(), 3, x.data_ptr() + 8) == _capi.CONV2D_EOVERLAP
    with pytest.raises(TypeError):
        pkg.conv2d_single(x.cpu(), f.cpu())  # no CPU fallback
    with pytest.raises(_capi.Conv2dError):
        pkg.conv2d_single(torch.zeros((2, 10), device=DEV), f)


# --------------------------------------------------------------------------------------------
# BASELINE.json configs at full size, EVERY output (configs[4]: every output of the band seams and of
# two whole bands), in the launch configuration bench.py times
# --------------------------------------------------------------------------------------------
@pytest.mark.parametrize("S", [1024, 2048, 4096, 8192])
def test_config1_sweep_full_size_every_output(cuda_device, S):
    """configs[1]: 1024^2..8192^2 x K in {3,..,15}, the bench launch configuration (one conv2d_single
    call per point on the current stream, automatic band height); every output against the oracle."""
    x = dev_image((S, S), "img", seed=synth.BASE_SEED + 1)
    xh = x.cpu().numpy()
    for K in (3, 5, 7, 9, 11, 13, 15):
        f = _filt(K, "rand", seed=synth.BASE_SEED + K)
        y = pkg.conv2d_single(x, f)
        torch.cuda.synchronize()
        check_full_single_host(xh, f.cpu().numpy(), y.cpu().numpy())
        del y


def test_config4_32768_k15_seams_and_bands(cuda_device):
    """configs[4]: one 32768^2 image, K=15 (4 GiB in + 4 GiB out) in one launch on one B200. Every
    output within K rows of each of the 7 seams of the 8-way row-band split (shard.row_band, the
    multi-GPU decomposition), plus every output of two whole bands (the first and the last), against
    the oracle; and each band computed on its own (what a rank computes) equals the one-launch rows
    bit for bit at the seams."""
    from paper_conf_cluster_luzw20_b200 import shard

    S, K = 32768, 15
    free, _ = torch.cuda.mem_get_info()
    if free < 10 * (1 << 30):
        pytest.skip("needs ~9 GiB of free HBM")
    x = dev_image((S, S), "img", seed=synth.BASE_SEED + 4)
    f = _filt(K, "gauss")
    fh = f.cpu().numpy()
    y = pkg.conv2d_single(x, f)
    torch.cuda.synchronize()
    Ho = S - K + 1
    bands = [shard.row_band(S, S, K, 8, r) for r in range(8)]

    def check_rows(o0, o1):
        xh = x[o0:o1 + K - 1].cpu().numpy()
        check_full_single_host(xh, fh, y[o0:o1].cpu().numpy())

    for b in bands[:-1]:  # seams: output rows [o1 - K, o1 + K) around each band end
        check_rows(max(0, b.o1 - K), min(Ho, b.o1 + K))
    for b in (bands[0], bands[-1]):  # two whole bands
        check_rows(b.o0, b.o1)
    for b in bands:  # a band computed alone (rows o0 .. o1+K-1) equals the one-launch rows
        lo, hi = b.o0, b.o1
        for a0, a1 in ((lo, min(hi, lo + 2 * K)), (max(lo, hi - 2 * K), hi)):
            part = pkg.conv2d_single(x[a0:a1 + K - 1], f)
            assert torch.equal(part, y[a0:a1]), (b.rank, a0, a1)


@pytest.mark.parametrize("variant", [1, 2, 3, 4, 5, 6, 7, 9, 13, 15, 20, 22, 23, 25, 26, 27, 40, 42, 43, 48, 49])
def test_every_kernel_variant_bitwise_equal(cuda_device, variant):
    """Every instantiation (filter in shared / constant memory, 1 or 2 column chunks -- the two-chunk
    ones with FFMA2 --, guarded or unguarded band prologue/epilogue, wide lanes 20-29, the slot-paired
    FFMA2 ring 48/49) of the one-warp-tile kernels gives the same bits as variant 1, and passes the
    oracle. (The default takes the filter-row split kernel for W <= 1024, K >= 11;
    its bits are covered by test_split_variants.)"""
    shapes = [(40, 300), (77, 1030), (300, 517)]
    try:
        for K in (1, 2, 3, 5, 8, 9, 12, 15):
            if ((variant == 13 and not 5 <= K <= 9) or (variant == 15 and K < 10)
                    or (variant in (48, 49) and (K % 2 == 0 or K < 3))):
                continue  # variants 13 / 15 / 48-49 exist for K = 5..9 / K >= 10 / odd K >= 3 only
            f = _filt(K, "rand", seed=K)
            for (dh, W) in shapes:
                x = dev_image((K + dh, W), "img", seed=K * 7 + W)
                _capi.debug_set_variant(1)
                ref = pkg.conv2d_single(x, f)
                _capi.debug_set_variant(variant)
                got = pkg.conv2d_single(x, f)
                torch.cuda.synchronize()
                assert torch.equal(got, ref), (variant, K, dh, W)
                if W == 300:
                    check_full_single(x, f, got)
                for bh in (1, 3, K + 1):
                    assert torch.equal(pkg.conv2d_single(x, f, band_h=bh), ref), (variant, K, bh)
    finally:
        _capi.debug_set_variant(0)


@pytest.mark.parametrize("K", [3, 4, 7, 11, 13, 15])
def test_split_variants(cuda_device, K):
    """Filter-row split kernel (conv2d_split.cuh): cluster of 2 one-warp CTAs (variant 10, the default
    for W <= 1024 and K >= 11), one CTA of 2 warps (11) and of 3 warps (12). Each passes the oracle on
    ragged / misaligned-pitch shapes, is bitwise band-independent (chunk tails, one-row bands), is
    exact on integer data, and 10 and 11 (same split, same sums) agree bit for bit."""
    shapes = [(1, 300), (40, 301), (77, 1030), (300, 517), (9, 129)]
    f = _filt(K, "rand", seed=K)
    try:
        for (dh, W) in shapes:
            x = dev_image((K + dh, W), "img", seed=K * 11 + W)
            outs = {}
            for v in (10, 11, 12):
                _capi.debug_set_variant(v)
                y = pkg.conv2d_single(x, f)
                torch.cuda.synchronize()
                check_full_single(x, f, y)
                for bh in (1, 5, 9, K + 2):
                    assert torch.equal(pkg.conv2d_single(x, f, band_h=bh), y), (v, K, W, bh)
                outs[v] = y
            assert torch.equal(outs[10], outs[11]), (K, dh, W)
            xi = dev_image((K + dh, W), "int", seed=K + W)
            fi = _filt(K, "int", seed=K)
            for v in (10, 12):
                _capi.debug_set_variant(v)
                check_full_single(xi, fi, pkg.conv2d_single(xi, fi), exact=True)
        _capi.debug_set_variant(0)
        if K >= 11:  # the default is variant 10 for narrow images
            x = dev_image((K + 50, 1000), "img", seed=K)
            y0 = pkg.conv2d_single(x, f)
            _capi.debug_set_variant(10)
            assert torch.equal(pkg.conv2d_single(x, f), y0)
    finally:
        _capi.debug_set_variant(0)


def test_cuda_graph_capture_and_replay(cuda_device):
    """Calls captured into a CUDA graph (shared-memory filter path) replay correctly, and filters
    updated between replays are picked up (the graph reads the filter tensor at replay time)."""
    x = dev_image((300, 700), "img")
    f = _filt(7)
    y = torch.empty((294, 694), device=DEV)
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        pkg.conv2d_single(x, f, out=y)  # warm-up outside capture
    torch.cuda.current_stream().wait_stream(s)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        pkg.conv2d_single(x, f, out=y)
    g.replay()
    torch.cuda.synchronize()
    check_full_single(x, f, y)
    f.copy_(_filt(7, "gauss"))
    x.copy_(dev_image((300, 700), "sym", seed=9))
    g.replay()
    torch.cuda.synchronize()
    check_full_single(x, f, y)


def test_concurrent_streams_different_filters(cuda_device):
    """Calls with the same K on two streams with different filters never see each other's filter
    (constant-slot reuse is ordered by events)."""
    x = dev_image((2000, 2048), "img")
    fs = [_filt(15, "rand", seed=s) for s in range(6)]
    outs = [torch.empty((1986, 2034), device=DEV) for _ in fs]
    streams = [torch.cuda.Stream() for _ in range(3)]
    for s in streams:
        s.wait_stream(torch.cuda.current_stream())
    for i, f in enumerate(fs):
        st = streams[i % 3]
        with torch.cuda.stream(st):
            pkg.conv2d_single(x, f, out=outs[i], stream=st)
    torch.cuda.synchronize()
    for f, y in zip(fs, outs):
        assert torch.equal(y, pkg.conv2d_single(x, f))


@pytest.mark.parametrize("pinned", [True, False])
def test_host_buffer_pipeline(cuda_device, pinned):
    """conv2d_single_host (H2D / kernel / D2H chunk pipeline) equals the device-resident call bit for
    bit, for chunk sizes that do and do not divide the output height."""
    for (H, W, K) in [(1000, 777, 3), (517, 1024, 15), (40, 300, 7)]:
        xh = synth.fill_np(H, synth.TAG_INPUT, (H, W), "img")
        fh = synth.make_filter(K, K, "rand")[0, 0]
        x = torch.from_numpy(xh)
        f = torch.from_numpy(fh)
        if pinned:
            x = x.pin_memory()
            f = f.pin_memory()
        ref = pkg.conv2d_single(x.cuda(), f.cuda()).cpu()
        for chunk in (0, 1, 7, 64, 10 ** 6):
            out = pkg.conv2d_single_host(x, f, chunk_rows=chunk)
            torch.cuda.synchronize()
            assert torch.equal(out, ref), (H, W, K, chunk)


@pytest.mark.parametrize("K", [1, 3, 7, 12, 15])
def test_halo_segment_bitwise(cuda_device, K):
    """conv2d_single_halo (row-band halo read in place): the rows of x followed by
    the rows of a SEPARATE allocation give the same bits as conv2d_single on the concatenation, for
    halo_rows 0..K-1 and more, narrow (split kernel) and wide images, aligned and misaligned halos."""
    f = _filt(K, "rand", seed=K)
    for (H, W) in [(40, 301), (K + 70, 1030), (200, 2052)]:
        full = dev_image((H + K + 3, W), "img", seed=K + W)
        for hr in sorted({0, 1, max(K - 1, 0), K + 3}):
            x = full[:H].clone()
            halo_store = torch.empty(((hr + 1) * W + 3,), device=DEV)
            for off in (0, 1):  # off=1: the halo rows start 4 bytes past a 16-byte boundary
                halo = halo_store[off:off + hr * W].view(hr, W)
                halo.copy_(full[H:H + hr])
                if H + hr < K:
                    continue
                ref = pkg.conv2d_single(full[:H + hr].contiguous(), f)
                got = pkg.conv2d_single_halo(x, halo, f)
                torch.cuda.synchronize()
                assert torch.equal(got, ref), (K, H, W, hr, off)
                if off == 1 and hr == max(K - 1, 0):  # the row-band case: every output vs the oracle
                    check_full_single(full[:H + hr], f, got)
    x = dev_image((30, 64), "img")
    halo = dev_image((K, 64), "img", seed=5)
    y = torch.empty((30 + K - K + 1, 64 - K + 1), device=DEV)
    assert _capi.conv2d_single_halo(x.data_ptr(), 30, 64, 0, 2, _filt(K).data_ptr(), K, y.data_ptr()) == \
        _capi.CONV2D_ENULL
    assert _capi.conv2d_single_halo(x.data_ptr(), 30, 64, halo.data_ptr(), -1, _filt(K).data_ptr(), K,
                                    y.data_ptr()) == _capi.CONV2D_ESHAPE
    assert _capi.conv2d_single_halo(x.data_ptr(), 30, 64, halo.data_ptr(), K, _filt(K).data_ptr(), K,
                                    halo.data_ptr()) == _capi.CONV2D_EOVERLAP


@pytest.mark.parametrize("K", [1, 3, 5, 7, 11, 15])
def test_single_batch_equals_per_image(cuda_device, K):
    """conv2d_single_batch (one launch over N images; the bench's sharding unit): bitwise equal to
    conv2d_single on every image, every output against the oracle, for small images (one wave holds
    all of them), narrow images with large K (filter-row split kernel), ragged and misaligned widths."""
    for (N, H, W) in [(5, K + 40, 300), (3, K + 90, 1030), (9, K + 7, 129), (2, 2 * K + 200, 1024), (1, K + 5, 77)]:
        x = dev_image((N, H, W), "img", seed=N * 100 + K)
        f = _filt(K, "rand", seed=K)
        y = pkg.conv2d_single_batch(x, f)
        torch.cuda.synchronize()
        for n in range(N):
            assert torch.equal(y[n], pkg.conv2d_single(x[n], f)), (K, N, H, W, n)
        xh, fh, yh = x.cpu().numpy(), f.cpu().numpy(), y.cpu().numpy()
        for n in range(N):
            check_full_single_host(xh[n], fh, yh[n])
    xi = dev_image((4, K + 30, 260), "int", seed=K)
    fi = _filt(K, "int", seed=K)
    yi = pkg.conv2d_single_batch(xi, fi)
    for n in range(4):
        check_full_single(xi[n], fi, yi[n], exact=True)


"""GPU parity of conv2d_multi (C ABI via the binding) against the CPU oracle: small shapes element by
element for every K, F not a multiple of the F-block, ragged widths; the BASELINE.json multi-channel
configs at full size, every output."""
import numpy as np
import pytest
import torch

import paper_conf_cluster_luzw20_b200 as pkg
from gen import synth
from tests.gpu_helpers import check_full_multi, check_full_single, dev_image

pytestmark = pytest.mark.gpu
DEV = "cuda"


def _w(F, C, K, dist="he", seed=5):
    return torch.from_numpy(synth.make_filter(seed, K, dist, F=F, C=C)).to(DEV)


@pytest.mark.parametrize("K", list(range(1, 16)))
def test_all_k_small(cuda_device, K):
    for (N, C, F, dh, dw) in [(1, 1, 1, 0, 0), (2, 3, 5, 7, 40), (1, 2, 9, 3, 131), (3, 1, 3, 20, 9)]:
        x = dev_image((N, C, K + dh, K + dw), "sym", seed=K + N)
        w = _w(F, C, K, seed=K)
        check_full_multi(x, w, pkg.conv2d_multi(x, w))


@pytest.mark.parametrize("K", [1, 3, 5, 7, 15])
def test_integer_bitwise(cuda_device, K):
    x = dev_image((2, 3, K + 17, 260), "int", seed=K)
    w = _w(7, 3, K, "int", seed=K)
    check_full_multi(x, w, pkg.conv2d_multi(x, w), exact=True)


def test_reduces_to_single(cuda_device):
    for K in (3, 7):
        x = dev_image((1, 1, 90, 300), "img", seed=K)
        w = _w(1, 1, K, "rand")
        ym = pkg.conv2d_multi(x, w)
        ys = pkg.conv2d_single(x[0, 0].contiguous(), w[0, 0].contiguous())
        check_full_single(x[0, 0], w[0, 0], ys)
        check_full_multi(x, w, ym)


def test_band_and_batch_split_bitwise(cuda_device):
    """Band height and batch sharding leave every output bit unchanged."""
    x = dev_image((6, 3, 70, 150), "img")
    w = _w(10, 3, 5)
    ref = pkg.conv2d_multi(x, w)
    for bh in (1, 3, 11, 1000):
        assert torch.equal(pkg.conv2d_multi(x, w, band_h=bh), ref)
    assert torch.equal(pkg.conv2d_multi(x[2:5].contiguous(), w), ref[2:5])
    assert torch.equal(pkg.conv2d_multi(x, w[3:8].contiguous()), ref[:, 3:8])


def test_config2_resnet_3x3(cuda_device):
    """configs[2]: N=32, C=F=64, 56x56, K=3 -- every output against the oracle."""
    N, C, F, S, K = 32, 64, 64, 56, 3
    x = dev_image((N, C, S, S), "sym", seed=synth.BASE_SEED + 2)
    w = _w(F, C, K, "he", seed=synth.BASE_SEED + 2)
    check_full_multi(x, w, pkg.conv2d_multi(x, w))


def test_config3_small_c_large_k(cuda_device):
    """configs[3]: N=128, C=3, F=64, 224x224, K=7 (R16: N=128) -- every output."""
    N, C, F, S, K = 128, 3, 64, 224, 7
    x = dev_image((N, C, S, S), "img", seed=synth.BASE_SEED + 3)
    w = _w(F, C, K, "he", seed=synth.BASE_SEED + 3)
    y = pkg.conv2d_multi(x, w)
    torch.cuda.synchronize()
    check_full_multi(x, w, y)


def test_config3_batch_shard_bitwise(cuda_device):
    """configs[3] batch-sharded as bench.py --gpus G shards it (shard.batch_range, 128/G images per
    rank): each shard computed alone equals the one-call rows bit for bit."""
    from paper_conf_cluster_luzw20_b200 import shard

    N, C, F, S, K = 128, 3, 64, 224, 7
    x = dev_image((N, C, S, S), "img", seed=synth.BASE_SEED + 3)
    w = _w(F, C, K, "he", seed=synth.BASE_SEED + 3)
    y = pkg.conv2d_multi(x, w)
    for G in (2, 8):
        for r in range(G):
            n0, n1 = shard.batch_range(N, G, r)
            assert torch.equal(pkg.conv2d_multi(x[n0:n1], w), y[n0:n1]), (G, r)


@pytest.mark.parametrize("layer", [("CONV1", 28, 128, 3), ("CONV3", 12, 64, 5), ("CONV4", 14, 16, 5),
                                   ("CONV10", 112, 128, 3)])
def test_table1_layers(cuda_device, layer):
    """PAPER.md Table I layer shapes at C in {1, 3}, reduced batch, every output."""
    name, S, F, K = layer
    for C in (1, 3):
        x = dev_image((4, C, S, S), "img", seed=S + C)
        w = _w(F, C, K, "he", seed=F)
        check_full_multi(x, w, pkg.conv2d_multi(x, w))


@pytest.mark.parametrize("shape", [(2, 64, 56, 56, 64, 3), (1, 3, 40, 45, 16, 5), (2, 16, 20, 37, 100, 3),
                                   (1, 8, 33, 30, 64, 7), (3, 1, 28, 28, 32, 3), (1, 4, 19, 21, 256, 1),
                                   (1, 3, 7, 7, 300, 7), (2, 2, 9, 130, 129, 2), (40, 3, 30, 33, 40, 3),
                                   (1, 1, 15, 15, 1, 15)])
def test_tensor_core_variant(cuda_device, shape):
    """conv2d_multi_tc (tcgen05 3xTF32 implicit GEMM) meets the same 1e-5*sum|x||w| acceptance."""
    N, C, H, W, F, K = shape
    x = dev_image((N, C, H, W), "sym", seed=C + F)
    w = _w(F, C, K, "he", seed=F)
    check_full_multi(x, w, pkg.conv2d_multi_tc(x, w))


def test_tensor_core_variant_config2(cuda_device):
    """configs[2] at full size through the tensor-core variant, every output."""
    N, C, F, S, K = 32, 64, 64, 56, 3
    x = dev_image((N, C, S, S), "sym", seed=synth.BASE_SEED + 2)
    w = _w(F, C, K, "he", seed=synth.BASE_SEED + 2)
    check_full_multi(x, w, pkg.conv2d_multi_tc(x, w))


@pytest.mark.parametrize("layer", [("CONV1", 28, 128, 3), ("CONV3", 12, 64, 5), ("CONV5", 24, 256, 5),
                                   ("CONV8", 28, 512, 3), ("CONV11", 224, 64, 3)])
def test_tensor_core_variant_table1(cuda_device, layer):
    """PAPER.md Table I layer shapes through the tensor-core variant, C in {1, 3},
    reduced batch, every output."""
    name, S, F, K = layer
    for C in (1, 3):
        x = dev_image((2, C, S, S), "img", seed=S + C)
        w = _w(F, C, K, "he", seed=F)
        check_full_multi(x, w, pkg.conv2d_multi_tc(x, w))


def test_tensor_core_variant_config3(cuda_device):
    """configs[3] (N=128, C=3, F=64, 224^2, K=7) at full size through the tensor-core variant, every
    output."""
    N, C, F, S, K = 128, 3, 64, 224, 7
    x = dev_image((N, C, S, S), "img", seed=synth.BASE_SEED + 3)
    w = _w(F, C, K, "he", seed=synth.BASE_SEED + 3)
    check_full_multi(x, w, pkg.conv2d_multi_tc(x, w))


@pytest.mark.parametrize("K", [1, 3, 5, 9, 15])
def test_eight_lane_segments(cuda_device, K):
    """8-lane segments (four images per warp, multi variant 7; the default for narrow layers): parity
    with N not a multiple of 4, widths past one 32-column segment, integer data exact, band-split bits."""
    from paper_conf_cluster_luzw20_b200 import _capi

    try:
        _capi.debug_set_multi_variant(7)
        for (N, C, F, dh, dw) in [(5, 3, 9, 5, 7), (4, 1, 17, 12, 30), (2, 2, 3, 3, 40), (9, 1, 8, 1, 0)]:
            x = dev_image((N, C, K + dh, K + dw), "img", seed=K + N)
            w = _w(F, C, K, seed=K + F)
            y = pkg.conv2d_multi(x, w)
            check_full_multi(x, w, y)
            for bh in (1, 4):
                assert torch.equal(pkg.conv2d_multi(x, w, band_h=bh), y), (K, N, bh)
        xi = dev_image((6, 3, K + 9, K + 20), "int", seed=K)
        wi = _w(7, 3, K, "int", seed=K)
        check_full_multi(xi, wi, pkg.conv2d_multi(xi, wi), exact=True)
    finally:
        _capi.debug_set_multi_variant(0)

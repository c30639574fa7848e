"""GPU parity of conv2d_single_rect (rectangular FH x FW filters) against the oracle:
every (FH, FW) in 1..15 x 1..15 on ragged / misaligned shapes element by element, integer data bitwise,
square filters equal to conv2d_single, a wide image spanning several 256-column tiles and bands."""
import numpy as np
import pytest
import torch

import oracle
import paper_conf_cluster_luzw20_b200 as pkg
from gen import synth
from paper_conf_cluster_luzw20_b200 import _capi
from tests.gpu_helpers import TOL, dev_image

pytestmark = pytest.mark.gpu
DEV = "cuda"


def _rect_filter(FH, FW, dist="rand", seed=1):
    rng = np.random.default_rng(seed * 100 + FH * 16 + FW)
    if dist == "int":
        return torch.from_numpy(rng.integers(-4, 5, (FH, FW)).astype(np.float32)).to(DEV)
    return torch.from_numpy(((2 * rng.random((FH, FW)) - 1) / max(FH, FW)).astype(np.float32)).to(DEV)


def _check(x, f, y, exact=False):
    ref, bound, _ = oracle.conv2d_single_rect(x.cpu().numpy(), f.cpu().numpy())
    got = y.cpu().numpy()
    assert got.shape == ref.shape
    bad = (got != ref) if exact else ~oracle.within_tolerance(got, ref, bound, TOL)
    assert not bad.any(), f"{int(bad.sum())} outputs off, first at {np.argwhere(bad)[:3].tolist()}"


@pytest.mark.parametrize("FH", list(range(1, 16)))
def test_every_fw(cuda_device, FH):
    for FW in range(1, 16):
        f = _rect_filter(FH, FW)
        for (H, W) in [(FH + 37, FW + 300), (FH, FW + 1), (FH + 5, 531)]:
            x = dev_image((H, W), "img", seed=H * 7 + W + FW)
            _check(x, f, pkg.conv2d_single_rect(x, f))


@pytest.mark.parametrize("FH,FW", [(1, 15), (15, 1), (3, 7), (7, 3), (2, 11), (13, 4)])
def test_integer_bitwise_and_wide_images(cuda_device, FH, FW):
    xi = dev_image((FH + 70, 1100), "int", seed=FH + FW)
    fi = _rect_filter(FH, FW, "int")
    _check(xi, fi, pkg.conv2d_single_rect(xi, fi), exact=True)
    x = dev_image((FH + 600, 2050), "img", seed=FH * FW)  # several 256-column tiles, ragged right edge, bands
    f = _rect_filter(FH, FW)
    _check(x, f, pkg.conv2d_single_rect(x, f))


def test_misaligned_and_square(cuda_device):
    FH, FW = 5, 9
    f = _rect_filter(FH, FW)
    buf = dev_image((70 * 301 + 4,), "img")
    x = buf[1:1 + 70 * 301].view(70, 301)  # 4 bytes past a 16-byte boundary: scalar path
    _check(x, f, pkg.conv2d_single_rect(x, f))
    for K in (3, 8):
        fs = torch.from_numpy(synth.make_filter(2, K, "rand")[0, 0]).to(DEV)
        xs = dev_image((K + 90, 777), "img", seed=K)
        assert torch.equal(pkg.conv2d_single_rect(xs, fs), pkg.conv2d_single(xs, fs))


def test_rect_error_codes(cuda_device):
    x = torch.zeros((10, 10), device=DEV)
    f = torch.zeros((3, 5), device=DEV)
    y = torch.zeros((8, 6), device=DEV)
    assert _capi.conv2d_single_rect(x.data_ptr(), 10, 10, f.data_ptr(), 3, 16, y.data_ptr()) == _capi.CONV2D_EK
    assert _capi.conv2d_single_rect(x.data_ptr(), 10, 10, f.data_ptr(), 0, 5, y.data_ptr()) == _capi.CONV2D_ESHAPE
    assert _capi.conv2d_single_rect(x.data_ptr(), 10, 4, f.data_ptr(), 3, 5, y.data_ptr()) == _capi.CONV2D_ESHAPE
    assert _capi.conv2d_single_rect(x.data_ptr(), 10, 10, f.data_ptr(), 3, 5, x.data_ptr() + 8) == \
        _capi.CONV2D_EOVERLAP

"""GPU parity of conv2d_single_pad ('same' zero / replicate padding, true
convolution) against the CPU oracle (oracle.conv2d_single_pad), and its bitwise identity with
conv2d_single on the padded image and the rotated filter (same kernels, data movement only)."""
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
MODES = [("valid", True), ("same_zero", False), ("same_zero", True), ("same_replicate", False),
         ("same_replicate", True)]


def _check(x, f, padding, flip, y, exact=False):
    ref, bound, _ = oracle.conv2d_single_pad(x.cpu().numpy(), f.cpu().numpy(), padding, flip)
    yh = y.cpu().numpy()
    assert yh.shape == ref.shape
    bad = (yh != ref) if exact else ~oracle.within_tolerance(yh, ref, bound, TOL)
    assert not bad.any(), (padding, flip, int(bad.sum()), np.argwhere(bad)[:3].tolist())


@pytest.mark.parametrize("K", [1, 2, 3, 4, 5, 7, 8, 11, 15])
def test_pad_modes_match_oracle(cuda_device, K):
    f = torch.from_numpy(synth.make_filter(K, K, "rand")[0, 0]).to(DEV)
    shapes = [(K + 40, 301), (K + 9, 1030), (3, 5), (1, 1), (2 * K + 1, 129)]
    for (H, W) in shapes:
        x = dev_image((H, W), "img", seed=H * 7 + K)
        for padding, flip in MODES:
            if padding == "valid" and (H < K or W < K):
                continue
            y = pkg.conv2d_single_pad(x, f, padding, flip)
            torch.cuda.synchronize()
            _check(x, f, padding, flip, y)


@pytest.mark.parametrize("K", [3, 6, 13])
def test_pad_integer_data_exact(cuda_device, K):
    f = torch.from_numpy(synth.make_filter(K, K, "int")[0, 0]).to(DEV)
    x = dev_image((K + 33, 517), "int", seed=K)
    for padding, flip in MODES:
        _check(x, f, padding, flip, pkg.conv2d_single_pad(x, f, padding, flip), exact=True)


@pytest.mark.parametrize("K", [2, 3, 5, 12, 15])
def test_pad_is_conv2d_single_of_padded_image_bitwise(cuda_device, K):
    """'same' = valid on the padded image, flip = rotated filter: interior launch + border strips give
    the bits of one one-tile-kernel call on the fully padded image (variant 1 as the reference: the
    default would take the filter-row split for narrow images with K >= 11)."""
    pt = (K - 1) // 2
    f = torch.from_numpy(synth.make_filter(K + 1, K, "rand")[0, 0]).to(DEV)
    for (H, W) in [(200, 333), (K + 60, 2048), (K - 1, 50), (7, K + 2)]:
        x = dev_image((H, W), "sym", seed=W + K)
        for mode in ("constant", "replicate"):
            xp = torch.nn.functional.pad(x[None, None], (pt, K - 1 - pt, pt, K - 1 - pt), mode=mode)[0, 0]
            for flip in (False, True):
                g = torch.flip(f, (0, 1)) if flip else f
                _capi.debug_set_variant(1)
                try:
                    ref = pkg.conv2d_single(xp.contiguous(), g.contiguous())
                finally:
                    _capi.debug_set_variant(0)
                got = pkg.conv2d_single_pad(x, f, "same_zero" if mode == "constant" else "same_replicate", flip)
                torch.cuda.synchronize()
                assert torch.equal(got, ref), (K, H, W, mode, flip)


def test_pad_in_cuda_graph_and_errors(cuda_device):
    K = 5
    x = dev_image((90, 140), "img")
    f = torch.from_numpy(synth.make_filter(2, K, "rand")[0, 0]).to(DEV)
    y = torch.empty((90, 140), device=DEV)
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        pkg.conv2d_single_pad(x, f, "same_replicate", True, out=y)
    torch.cuda.current_stream().wait_stream(s)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        pkg.conv2d_single_pad(x, f, "same_replicate", True, out=y)
    y.zero_()
    g.replay()
    torch.cuda.synchronize()
    _check(x, f, "same_replicate", True, y)
    L = _capi.load()
    assert L.conv2d_single_pad(x.data_ptr(), 90, 140, f.data_ptr(), K, 3, y.data_ptr(), 0) == _capi.CONV2D_ESHAPE
    assert L.conv2d_single_pad(x.data_ptr(), 90, 140, f.data_ptr(), K, 8, y.data_ptr(), 0) == _capi.CONV2D_ESHAPE
    assert L.conv2d_single_pad(x.data_ptr(), 90, 140, f.data_ptr(), 16, 1, y.data_ptr(), 0) == _capi.CONV2D_EK
    assert L.conv2d_single_pad(x.data_ptr(), 3, 3, f.data_ptr(), K, 4, y.data_ptr(), 0) == _capi.CONV2D_ESHAPE
    assert L.conv2d_single_pad(x.data_ptr(), 90, 140, f.data_ptr(), K, 1, x.data_ptr(), 0) == _capi.CONV2D_EOVERLAP

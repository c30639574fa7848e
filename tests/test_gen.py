"""The shared seeded generator: numpy and torch implementations are bit-identical, shard-independent,
and produce the documented ranges."""
import numpy as np
import pytest
import torch

from gen import synth


def test_splitmix64_reference_vector():
    # First output of the published splitmix64 generator seeded with 0 (Vigna's reference code).
    assert int(synth.splitmix64_np(np.array([0], np.uint64))[0]) == 0xE220A8397B1DCDAF


@pytest.mark.parametrize("dist", synth.IMAGE_DISTS)
def test_numpy_torch_bit_identical(dist):
    a = synth.fill_np(123, synth.TAG_INPUT, (77, 129), dist, start=999)
    b = synth.fill_torch(123, synth.TAG_INPUT, (77, 129), dist, start=999).numpy()
    assert np.array_equal(a.view(np.uint32), b.view(np.uint32))


@pytest.mark.parametrize("dist", synth.IMAGE_DISTS)
def test_shard_independent(dist):
    full = synth.fill_np(5, 1, (40, 50), dist)
    top = synth.fill_np(5, 1, (17, 50), dist, start=0)
    bot = synth.fill_np(5, 1, (23, 50), dist, start=17 * 50)
    assert np.array_equal(full, np.concatenate([top, bot]))
    # chunked generation is the same as one shot
    assert np.array_equal(full, synth.fill_np(5, 1, (40, 50), dist, chunk=333))


def test_ranges_and_exactness():
    img = synth.fill_np(1, 1, (1 << 16,), "img")
    assert img.min() >= 0 and img.max() < 1
    assert np.all(img * 2 ** 24 == np.round(img * 2 ** 24))  # 24-bit dyadics, exact in fp32
    sym = synth.fill_np(1, 1, (1 << 16,), "sym")
    assert sym.min() >= -1 and sym.max() < 1 and abs(sym.mean()) < 0.02
    ints = synth.fill_np(1, 1, (1 << 16,), "int")
    assert set(np.unique(ints)) == set(range(-8, 9))


def test_filters():
    for K in (1, 3, 4, 15):
        g = synth.make_filter(0, K, "gauss")
        assert g.shape == (1, 1, K, K) and abs(float(g.astype(np.float64).sum()) - 1) < 1e-6
        d = synth.make_filter(0, K, "delta")
        assert d.sum() == 1 and d[0, 0, K // 2, K // 2] == 1
        b = synth.make_filter(0, K, "box")
        assert (b == 1).all()
        r = synth.make_filter(0, K, "rand")
        assert np.abs(r).max() <= 1.0 / K
        i = synth.make_filter(0, K, "int", F=2, C=3)
        assert i.shape == (2, 3, K, K) and np.abs(i).max() <= 4
    he = synth.make_filter(3, 7, "he", F=64, C=3)
    assert abs(he.std() - np.sqrt(2 / (3 * 49))) < 0.02 * np.sqrt(2 / (3 * 49)) * 5

"""SASS evidence checks of the built product library (CPU only: cuobjdump, no GPU).

The paper's dynamic->static index transformation exists to keep the per-thread
window (iTemp) and the output accumulators (Out) in registers: a kernel that spills them to local
memory has lost exactly what the method is about. Every kernel shipped in libconv2d.so must therefore
be free of LDL/STL, and the single-channel kernels must show the method's instruction signature:
FFMA / FFMA2 for row reuse and SHFL for column reuse; the multi-channel kernels FFMA2 over filter pairs."""
import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.path.join(ROOT, "tools"))


@pytest.fixture(scope="module")
def product_kernels():
    from paper_conf_cluster_luzw20_b200 import _build

    _build.build()
    import sass_report

    return sass_report.kernels(sass_report.LIBS["product"])


def test_no_spills_in_any_product_kernel(product_kernels):
    bad = {k: (c["LDL"], c["STL"]) for k, c in product_kernels.items() if c["LDL"] or c["STL"]}
    assert not bad, f"kernels with local-memory spills: {bad}"


def test_single_channel_kernels_carry_column_and_row_reuse(product_kernels):
    singles = {k: c for k, c in product_kernels.items() if "k_conv2d_single" in k or "k_conv2d_split" in k}
    assert singles
    for k, c in singles.items():
        assert c["FFMA"] + c["FFMA2"] > 0, k  # row reuse: FMA chains (scalar, or paired fma.rn.f32x2)
        kk = int(k.split("ILi", 1)[1].split("E", 1)[0])  # K, the first template argument
        if kk > 1:
            assert c["SHFL"] > 0, k  # column reuse: halo columns by warp shuffle, not reloads


def test_tensor_core_variant_uses_tcgen05(product_kernels):
    tc = {k: c for k, c in product_kernels.items() if "k_conv2d_multi_tc" in k}
    assert tc
    for k, c in tc.items():
        assert c["UTCHMMA"] + c["UTCQMMA"] > 0 and c["LDTM"] > 0, k


def test_multi_channel_kernels_pair_filters_and_shuffle(product_kernels):
    """The filter-blocked multi-channel kernel (conv2d_mob.cuh): paired FMAs over filter pairs, broadcast
    LDS of the staged F-block, SHFL for the column-reuse halo (K > 1)."""
    mob = {k: c for k, c in product_kernels.items() if "k_conv2d_mob" in k}
    assert mob
    for k, c in mob.items():
        assert c["FFMA2"] > 0 and c["LDS"] > 0, k
        kk = int(k.split("ILi", 1)[1].split("E", 1)[0])
        if kk > 1:
            assert c["SHFL"] > 0, k

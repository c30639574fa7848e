"""B200-native (sm_100a) direct fp32 convolution with the column and row reuse of Lu, Zhang & Wang,
"Optimizing GPU Memory Transactions for Convolution Operations" (IEEE Cluster 2020).

The product is libconv2d.so (C ABI, include/conv2d.h). This package is its thin Python binding:
    _capi   ctypes marshalling of the C entry points (same names)
    api     torch-tensor wrappers (device memory / streams only)
    shard   multi-GPU partitioning: batch, filter and row-band (a (K-1)-row halo by NCCL P2P, or read
            in place from the neighbour's memory over NVLink by conv2d_single_halo; symmetric
            memory or CUDA IPC mappings)
"""
from . import _capi
from .api import (conv2d_multi, conv2d_multi_host, conv2d_multi_tc, conv2d_single, conv2d_single_batch,
                  conv2d_single_direct, conv2d_single_rect, conv2d_single_halo, conv2d_single_host, conv2d_single_pad)

__all__ = ["_capi", "conv2d_multi", "conv2d_multi_host", "conv2d_multi_tc", "conv2d_single",
           "conv2d_single_batch", "conv2d_single_direct", "conv2d_single_rect", "conv2d_single_halo", "conv2d_single_host",
           "conv2d_single_pad"]

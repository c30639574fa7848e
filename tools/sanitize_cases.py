#!/usr/bin/env python
"""Small invocations of every product kernel family for compute-sanitizer (memcheck / racecheck /
initcheck): wide-lane and one-chunk single-channel kernels (register and cp.async-ring row fetch, shared
and constant filters), the filter-row split kernel (cluster of 2 CTAs, DSMEM), batches, the halo and
'same'-padding paths, rectangular filters, the multi-channel kernels (filter-blocked default at 4/8/16-lane
segments, FB = 8 / 4, misaligned input, large-C fallbacks) and the tcgen05 tensor-core variant, the host-buffer pipeline.

    compute-sanitizer --tool memcheck python tools/sanitize_cases.py
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402


def img(shape, seed=1):
    return synth.fill_torch(seed, 1, shape, "img", device="cuda")


def filt(K, seed=2):
    return torch.from_numpy(synth.make_filter(seed, K, "rand")[0, 0]).cuda()


def main():
    for K in (3, 5, 7, 11, 15):
        pkg.conv2d_single(img((K + 40, 8200)), filt(K))          # wide image: constant slot, wide / ring kernels
        pkg.conv2d_single(img((K + 30, 1000)), filt(K))          # narrow: smem filter / split kernel (K >= 11)
        pkg.conv2d_single(img((K + 21, 517)), filt(K))           # ragged right edge
        b = img(((K + 20) * 300 + 4,))
        pkg.conv2d_single(b[1:1 + (K + 20) * 300].view(K + 20, 300), filt(K))  # misaligned rows
        pkg.conv2d_single_batch(img((3, K + 17, 700)), filt(K))
        pkg.conv2d_single_halo(img((40, 600)), img((K - 1, 600), 3), filt(K))
        pkg.conv2d_single_pad(img((50, 260)), filt(K), "same_replicate", flip=True)
        pkg.conv2d_single_rect(img((K + 30, 530)), torch.rand((K, max(1, K - 2)), device="cuda"))
    # multi-channel: the filter-blocked kernel at 4/8/16-lane segments, FB = 8 and 4, the K <= 4 L1-prefetch
    # form, odd output pitch, the large-C fallbacks (FB = 4, then the one-filter round-1 kernel)
    for (N, C, H, W, F, K) in [(4, 3, 30, 33, 16, 3), (2, 64, 20, 20, 64, 3), (1, 3, 40, 260, 8, 7),
                               (5, 1, 28, 28, 20, 5), (2, 2, 19, 23, 3, 15), (3, 3, 20, 224, 24, 7),
                               (4, 8, 14, 56, 16, 3), (2, 3, 12, 29, 9, 5), (1, 40, 20, 60, 5, 15),
                               (1, 200, 18, 40, 3, 15)]:
        x = img((N, C, H, W))
        w = torch.from_numpy(synth.make_filter(4, K, "he", F=F, C=C)).cuda()
        pkg.conv2d_multi(x, w)
        if C * K * K <= (1 << 14):  # the tensor-core variant's im2col offset table bound (conv2d.h)
            pkg.conv2d_multi_tc(x, w)
        xb = img((N * C * H * W + 1,))[1:].view(N, C, H, W)  # misaligned input
        pkg.conv2d_multi(xb, w)
    xh = torch.rand((70, 300)).pin_memory()
    pkg.conv2d_single_host(xh, torch.rand((5, 5)), chunk_rows=16)
    torch.cuda.synchronize()
    print("sanitize cases: ok")


if __name__ == "__main__":
    main()

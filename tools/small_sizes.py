#!/usr/bin/env python
"""Per-call time of small single-channel convolutions (latency regime), per variant."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from paper_conf_cluster_luzw20_b200 import _capi  # noqa: E402


def per_call_us(fn, n=200):
    for _ in range(10):
        fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(n):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / n * 1e3


def main():
    variants = [int(v) for v in (sys.argv[1] if len(sys.argv) > 1 else "1,2,3,4").split(",")]
    for S in (16, 256, 1024, 2048):
        x = synth.fill_torch(1, 1, (S, S), "img", device="cuda")
        for K in (3, 9, 15):
            f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
            y = torch.empty((S - K + 1, S - K + 1), device="cuda")
            line = f"{S:5d}^2 K={K:2d}:"
            for v in variants:
                _capi.debug_set_variant(v)
                us = per_call_us(lambda: pkg.conv2d_single(x, f, out=y))
                line += f"  v{v} {us:7.2f} us"
            _capi.debug_set_variant(0)
            print(line, flush=True)


if __name__ == "__main__":
    main()

#!/usr/bin/env python
"""GPU-side time per call of back-to-back small conv2d_single calls: the stream is first blocked by
a long spin kernel (torch.cuda._sleep) while the host enqueues every call, so the events measure the
device timeline only (kernel + filter staging copy + launch gaps), not the host's issue rate.

    python tools/gpu_side_calls.py [--variants 0,1,2] [--n 100]
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from paper_conf_cluster_luzw20_b200 import _capi  # noqa: E402


def gpu_us(fn, n):
    for _ in range(5):
        fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda._sleep(int(2e8))  # ~100 ms of spinning: the host enqueues all n calls meanwhile
    e0.record()
    for _ in range(n):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / n * 1e3


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--variants", default="0,1,2")
    ap.add_argument("--n", type=int, default=100)
    a = ap.parse_args()
    for S in (64, 256, 1024, 2048):
        x = synth.fill_torch(1, 1, (S, S), "img", device="cuda")
        for K in (3, 7, 15):
            f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
            y = torch.empty((S - K + 1, S - K + 1), device="cuda")
            line = f"{S:5d}^2 K={K:2d}:"
            for v in [int(t) for t in a.variants.split(",")]:
                _capi.debug_set_variant(v)
                line += f"  v{v} {gpu_us(lambda: pkg.conv2d_single(x, f, out=y), a.n):7.2f} us"
            _capi.debug_set_variant(0)
            print(line, flush=True)


if __name__ == "__main__":
    main()

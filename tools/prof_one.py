#!/usr/bin/env python
"""Run one convolution a few times (for ncu captures and quick timing).

    python tools/prof_one.py single 8192 15 [--reps 3] [--direct] [--band BH]
    python tools/prof_one.py multi 32,64,56,56,64 3
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("kind", choices=["single", "multi"])
    ap.add_argument("shape")
    ap.add_argument("K", type=int)
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--direct", action="store_true")
    ap.add_argument("--band", type=int, default=0)
    ap.add_argument("--time", action="store_true")
    ap.add_argument("--variant", type=int, default=0)
    ap.add_argument("--mvariant", type=int, default=0)
    ap.add_argument("--tc", action="store_true", help="multi: the tensor-core variant conv2d_multi_tc")
    ap.add_argument("--batch", type=int, default=1, help="single: images per call (conv2d_single_batch)")
    a = ap.parse_args()
    pkg._capi.debug_set_variant(a.variant)
    pkg._capi.debug_set_multi_variant(a.mvariant)
    dev = torch.device("cuda")
    if a.kind == "single":
        S = [int(v) for v in a.shape.split(",")]
        H, W = (S[0], S[0]) if len(S) == 1 else S
        x = synth.fill_torch(1, 1, (a.batch, H, W), "img", device=dev)
        f = torch.from_numpy(synth.make_filter(1, a.K, "rand")[0, 0]).to(dev)
        if a.direct:
            fn = lambda: pkg.conv2d_single_direct(x[0], f)  # noqa: E731
        elif a.batch > 1:
            fn = lambda: pkg.conv2d_single_batch(x, f)  # noqa: E731
        else:
            fn = lambda: pkg.conv2d_single(x[0], f, band_h=a.band)  # noqa: E731
        px = (H - a.K + 1) * (W - a.K + 1) * a.batch
        work = px
    else:
        N, C, H, W, F = [int(v) for v in a.shape.split(",")]
        x = synth.fill_torch(1, 1, (N, C, H, W), "img", device=dev)
        w = torch.from_numpy(synth.make_filter(1, a.K, "he", F=F, C=C)).to(dev)
        fn = (lambda: pkg.conv2d_multi_tc(x, w)) if a.tc else (lambda: pkg.conv2d_multi(x, w, band_h=a.band))
        work = 2.0 * N * F * (H - a.K + 1) * (W - a.K + 1) * C * a.K * a.K
    for _ in range(a.reps):
        fn()
    torch.cuda.synchronize()
    if a.time:
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        n = 20
        e0.record()
        for _ in range(n):
            fn()
        e1.record()
        torch.cuda.synchronize()
        ms = e0.elapsed_time(e1) / n
        print(f"{a.kind} {a.shape} K={a.K}: {ms:.4f} ms/call, {work / ms / 1e6:.1f} G{'px' if a.kind == 'single' else 'FLOP'}/s")


if __name__ == "__main__":
    main()

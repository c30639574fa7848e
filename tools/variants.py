#!/usr/bin/env python
"""Time every single-channel kernel variant on the sweep points; check they agree bit for bit.

    python tools/variants.py [--sizes 8192,4096] [--ks 3,5,7,9,11,13,15] [--variants 1,2,3,4]
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


def time_call(fn, n=10):
    flush = torch.empty(256 << 20, dtype=torch.uint8, device="cuda")
    ts = []
    for _ in range(n):
        flush.zero_()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        fn()
        e1.record()
        torch.cuda.synchronize()
        ts.append(e0.elapsed_time(e1))
    ts.sort()
    return ts[len(ts) // 2]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sizes", default="8192,4096")
    ap.add_argument("--ks", default="3,5,7,9,11,13,15")
    ap.add_argument("--variants", default="1,2,3,4")
    ap.add_argument("--band", type=int, default=0)
    ap.add_argument("--minband", type=int, default=0)
    ap.add_argument("--batch", type=int, default=1, help="images per call (conv2d_single_batch when > 1)")
    a = ap.parse_args()
    _capi.debug_set_min_band(a.minband)
    for S in [int(v) for v in a.sizes.split(",")]:
        B = a.batch
        x = synth.fill_torch(1, 1, (B, S, S), "img", device="cuda")

        def call(x, f, out=None, band_h=0):
            if B == 1:
                return pkg.conv2d_single(x[0], f, out=None if out is None else out[0], band_h=band_h)[None]
            return pkg.conv2d_single_batch(x, f, out=out)
        for K in [int(v) for v in a.ks.split(",")]:
            f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
            ref = None
            line = f"{S}^2 K={K:2d}:"
            for v in [int(t) for t in a.variants.split(",")]:
                _capi.debug_set_variant(v)
                y = call(x, f, band_h=a.band)
                torch.cuda.synchronize()
                if ref is None:
                    ref = y.clone()
                same = torch.equal(y, ref)
                ms = time_call(lambda: call(x, f, out=y, band_h=a.band))
                px = (S - K + 1) ** 2 * B
                line += f"  v{v} {px / ms / 1e6:7.1f} Gpx/s ({2 * px * K * K / ms / 1e9:5.1f} TF){'' if same else ' MISMATCH'}"
            _capi.debug_set_variant(0)
            print(line, flush=True)


if __name__ == "__main__":
    main()

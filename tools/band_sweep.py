#!/usr/bin/env python
"""Band-height sweep of the default single-channel kernel: taller bands mean fewer resident warps but
less Alg. 2 case-1/3 (halo-row) work per output; prints Gpx/s per band height, bits checked.

    python tools/band_sweep.py [--sizes 1024,2048,4096] [--ks 3,7,11,15] [--mults 1,1.5,2,3,4]
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
from variants import time_call  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sizes", default="1024,2048,4096")
    ap.add_argument("--ks", default="3,5,7,9,11,13,15")
    ap.add_argument("--bands", default="0,8,16,24,32,48,64,96,128,192,256")
    ap.add_argument("--variant", type=int, default=0)
    a = ap.parse_args()
    _capi.debug_set_variant(a.variant)
    for S in [int(v) for v in a.sizes.split(",")]:
        x = synth.fill_torch(1, 1, (S, S), "img", device="cuda")
        for K in [int(v) for v in a.ks.split(",")]:
            f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
            ref = pkg.conv2d_single(x, f)
            torch.cuda.synchronize()
            px = (S - K + 1) ** 2
            line = f"{S}^2 K={K:2d}:"
            for b in [int(t) for t in a.bands.split(",")]:
                if b and b < K - 1:
                    continue
                y = pkg.conv2d_single(x, f, band_h=b)
                same = torch.equal(y, ref)
                ms = time_call(lambda: pkg.conv2d_single(x, f, out=y, band_h=b))
                line += f"  b{b}:{px / ms / 1e6:6.1f}{'' if same else '!'}"
            print(line, flush=True)


if __name__ == "__main__":
    main()

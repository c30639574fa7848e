#!/usr/bin/env python
"""Time single-channel variants (default, cluster filter-row split 10-14) per point; outputs checked
against the default variant (max |d| / max |ref|, must stay ~1e-7: the split only regroups sums).

    python tools/split_sweep.py [--sizes 256,1024,2048,4096,8192] [--ks 3,...,15] [--variants 0,10,...]
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))

import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from paper_conf_cluster_luzw20_b200 import _capi  # noqa: E402
from variants import time_call  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sizes", default="256,1024,2048,4096,8192")
    ap.add_argument("--ks", default="3,5,7,9,11,13,15")
    ap.add_argument("--variants", default="0,10,11,12,13,14")
    ap.add_argument("--minband", type=int, default=0)
    a = ap.parse_args()
    _capi.debug_set_min_band(a.minband)
    for S in [int(v) for v in a.sizes.split(",")]:
        x = synth.fill_torch(1, 1, (S, S), "img", device="cuda")
        for K in [int(v) for v in a.ks.split(",")]:
            f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
            _capi.debug_set_variant(0)
            ref = pkg.conv2d_single(x, f)
            torch.cuda.synchronize()
            scale = float(ref.abs().max())
            px = (S - K + 1) ** 2
            line = f"{S}^2 K={K:2d}:"
            for v in [int(t) for t in a.variants.split(",")]:
                _capi.debug_set_variant(v)
                try:
                    y = pkg.conv2d_single(x, f)
                    torch.cuda.synchronize()
                except Exception as e:  # noqa: BLE001
                    line += f"  v{v} err({e})"
                    continue
                err = float((y - ref).abs().max()) / scale
                ms = time_call(lambda: pkg.conv2d_single(x, f, out=y))
                line += f"  v{v} {px / ms / 1e6:6.1f}{'' if err < 1e-6 else f' ERR{err:.1e}'}"
            _capi.debug_set_variant(0)
            print(line, flush=True)


if __name__ == "__main__":
    main()

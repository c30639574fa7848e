#!/usr/bin/env python
"""Back-to-back per-call device time (us) of conv2d_single per variant at mid sizes: the constant-slot
default (staging copy + events per call) against the shared-memory filter variants (no staging)."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from paper_conf_cluster_luzw20_b200 import _capi  # noqa: E402
from small_sizes import per_call_us  # noqa: E402


def main():
    variants = [int(v) for v in (sys.argv[1] if len(sys.argv) > 1 else "0,1,2").split(",")]
    for S in (512, 1024, 2048, 4096):
        # several distinct images so the back-to-back calls do not all hit L2
        xs = [synth.fill_torch(i, 1, (S, S), "img", device="cuda") for i in range(max(1, 8 * 2048 // S))]
        for K in (3, 5, 7, 9, 11):
            f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
            ys = [torch.empty((S - K + 1, S - K + 1), device="cuda") for _ in xs]
            line = f"{S:5d}^2 K={K:2d}:"
            for v in variants:
                _capi.debug_set_variant(v)
                it = [0]

                def call():
                    i = it[0] % len(xs)
                    it[0] += 1
                    pkg.conv2d_single(xs[i], f, out=ys[i])
                us = per_call_us(call, n=100)
                line += f"  v{v} {us:8.2f}"
            _capi.debug_set_variant(0)
            print(line, flush=True)


if __name__ == "__main__":
    main()

#!/usr/bin/env python
"""'same'-padding call (conv2d_single_pad) vs the valid call at 8192^2 K = 3/5/7 across single-channel
kernel variants (tuning build): us per call, bits checked across variants.

    python tools/pad_variants.py
"""
import sys, torch
import os
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT); sys.path.insert(0, os.path.join(ROOT, 'tools'))
import paper_conf_cluster_luzw20_b200 as pkg
from paper_conf_cluster_luzw20_b200 import _capi
from gen import synth
from variants import time_call
x = synth.fill_torch(1, 1, (8192, 8192), "img", device="cuda")
for K in (3, 5, 7):
    f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
    line = f"K={K}:"
    ref = None
    for v in (0, 3, 4, 17, 18, 20, 23, 27):
        _capi.debug_set_variant(v)
        try:
            y = pkg.conv2d_single_pad(x, f, "same_zero")
            torch.cuda.synchronize()
        except Exception as e:
            line += f" v{v} n/a"; continue
        if ref is None: ref = y.clone()
        ms = time_call(lambda: pkg.conv2d_single_pad(x, f, "same_zero"))
        ms_valid = time_call(lambda: pkg.conv2d_single(x, f))
        line += f" v{v} {ms*1e3:.0f}us/{ms_valid*1e3:.0f}us{'' if torch.equal(y, ref) else '!'}"
    _capi.debug_set_variant(0)
    print(line, flush=True)

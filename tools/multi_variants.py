#!/usr/bin/env python
"""Time the multi-channel kernel variants on the BASELINE configs and Table I layers; check bits.

    python tools/multi_variants.py [--variants 0,1,2,3,4,9]
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

SHAPES = {  # name: (N, C, H, W, F, K)
    "config2 N32 C64 56^2 F64 K3": (32, 64, 56, 56, 64, 3),
    "config3 N128 C3 224^2 F64 K7": (128, 3, 224, 224, 64, 7),
    "TableI CONV1 C3": (128, 3, 28, 28, 128, 3),
    "TableI CONV2 C3": (128, 3, 56, 56, 64, 3),
    "TableI CONV5 C3": (128, 3, 24, 24, 256, 5),
    "TableI CONV9 C3": (128, 3, 56, 56, 256, 3),
    "TableI CONV11 C1": (128, 1, 224, 224, 64, 3),
}
TABLE1 = [("CONV1", 28, 128, 3), ("CONV2", 56, 64, 3), ("CONV3", 12, 64, 5), ("CONV4", 14, 16, 5),
          ("CONV5", 24, 256, 5), ("CONV6", 24, 64, 5), ("CONV7", 28, 16, 5), ("CONV8", 28, 512, 3),
          ("CONV9", 56, 256, 3), ("CONV10", 112, 128, 3), ("CONV11", 224, 64, 3)]


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
    ap.add_argument("--variants", default="0,1,2,3,4,9")
    ap.add_argument("--only", default="")
    ap.add_argument("--table1", action="store_true", help="all 22 Table I layers (C in {1, 3}) + the two configs")
    a = ap.parse_args()
    shapes = dict(SHAPES)
    if a.table1:
        shapes = {k: v for k, v in SHAPES.items() if k.startswith("config")}
        for C in (1, 3):
            for nm, S, F, K in TABLE1:
                shapes[f"TableI {nm} C{C}"] = (128, C, S, S, F, K)
    for name, (N, C, H, W, F, K) in shapes.items():
        if a.only and a.only not in name:
            continue
        x = synth.fill_torch(1, 1, (N, C, H, W), "img", device="cuda")
        w = torch.from_numpy(synth.make_filter(1, K, "he", F=F, C=C)).cuda()
        flops = 2.0 * N * F * (H - K + 1) * (W - K + 1) * C * K * K
        ref = None
        line = f"{name:32s}"
        for vs in a.variants.split(","):
            # "tc" = tensor-core variant (default tuning), "tcNN" = with multi variant override NN
            v = -1 if vs.startswith("tc") else int(vs)
            fn = (lambda out=None: pkg.conv2d_multi_tc(x, w, out=out)) if v < 0 else \
                (lambda out=None: pkg.conv2d_multi(x, w, out=out))
            _capi.debug_set_multi_variant(int(vs[2:] or 0) if v < 0 else v)
            try:
                y = fn()
                torch.cuda.synchronize()
            except Exception as e:  # variant not applicable
                line += f"  v{v} n/a({type(e).__name__})"
                continue
            if ref is None:
                ref = y.clone()
            same = torch.equal(y, ref)
            ms = time_call(lambda: fn(out=y))
            if v < 0:  # the tensor-core variant is not bitwise equal: report its max relative deviation
                dev = float(((y - ref).abs().max() / ref.abs().max().clamp_min(1e-30)).item())
                line += f"  {vs} {flops / ms / 1e9:6.1f} TF (max dev {dev:.1e})"
            else:
                line += f"  v{v} {flops / ms / 1e9:6.1f} TF{'' if same else ' DIFF'}"
        _capi.debug_set_multi_variant(0)
        print(line, flush=True)


if __name__ == "__main__":
    main()

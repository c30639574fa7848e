#!/usr/bin/env python
"""Device latency of ONE small conv2d_single call (events around a single launch on an idle GPU, after
an L2-flushing write), per variant and band height: the configs[0] regime."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from paper_conf_cluster_luzw20_b200 import _capi  # noqa: E402


def lat_us(fn, graph, n=50):
    flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
    g = None
    if graph:
        s = torch.cuda.Stream()
        s.wait_stream(torch.cuda.current_stream())
        with torch.cuda.stream(s):
            fn()
        torch.cuda.current_stream().wait_stream(s)
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g):
            fn()
    ts = []
    for _ in range(n):
        flush.zero_()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        torch.cuda.synchronize()
        e0.record()
        g.replay() if g is not None else fn()
        e1.record()
        torch.cuda.synchronize()
        ts.append(e0.elapsed_time(e1) * 1e3)
    ts.sort()
    return ts[len(ts) // 2]


def main():
    for S, K in ((256, 3), (256, 9), (256, 15), (512, 3)):
        x = synth.fill_torch(1, 1, (S, S), "img", device="cuda")
        f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
        y = torch.empty((S - K + 1, S - K + 1), device="cuda")
        line = f"{S}^2 K={K:2d}:"
        for v in (0, 1, 2, 7, 9):
            for bh in (0, 1, 2, 8):
                _capi.debug_set_variant(v)
                try:
                    us = lat_us(lambda: pkg.conv2d_single(x, f, out=y, band_h=bh), graph=(v in (0, 1, 2)))
                    line += f"  v{v}b{bh} {us:5.1f}"
                except Exception:  # noqa: BLE001
                    line += f"  v{v}b{bh} err"
        _capi.debug_set_variant(0)
        print(line, flush=True)


if __name__ == "__main__":
    main()

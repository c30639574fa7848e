#!/usr/bin/env python
"""Per-step end-to-end times (conv2d_single_host over the sweep), to see their spread."""
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402

sizes = (8192, 4096, 2048, 1024)
ks = (3, 5, 7, 9, 11, 13, 15)
pts = []
for S in sizes:
    for K in ks:
        x = synth.fill_torch(1, 1, (S, S), "img").pin_memory()
        f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).pin_memory()
        y = torch.empty((S - K + 1, S - K + 1), pin_memory=True)
        pts.append((x, f, y))
streams = [torch.cuda.Stream() for _ in range(2)]
main = torch.cuda.current_stream()
mode = sys.argv[1] if len(sys.argv) > 1 else "host"


def one():
    for s in streams:
        s.wait_stream(main)
    for i, (x, f, y) in enumerate(pts):
        pkg.conv2d_single_host(x, f, stream=streams[i % 2], out_host=y)
    for s in streams:
        main.wait_stream(s)


for it in range(8):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    one()
    e1.record()
    torch.cuda.synchronize()
    print(f"step {it}: {e0.elapsed_time(e1):.1f} ms (wall {1e3 * (time.perf_counter() - t0):.1f})", flush=True)

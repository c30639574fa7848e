#!/usr/bin/env python
"""Host-side cost per call of the small-image path (latency regime): the Python API, the raw C ABI
call, and the C ABI with the shared-memory filter variant (no constant-slot staging), against a
plain torch launch for scale. Prints host us/call (enqueue rate) and device us/call (events)."""
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from paper_conf_cluster_luzw20_b200 import _capi  # noqa: E402


def measure(fn, n=2000):
    for _ in range(50):
        fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    t0 = time.perf_counter()
    e0.record()
    for _ in range(n):
        fn()
    e1.record()
    t1 = time.perf_counter()
    torch.cuda.synchronize()
    return (t1 - t0) / n * 1e6, e0.elapsed_time(e1) / n * 1e3


def main():
    L = _capi.load()
    for S, K in ((16, 3), (256, 3), (256, 15), (1024, 3)):
        x = synth.fill_torch(1, 1, (S, S), "img", device="cuda")
        f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
        y = torch.empty((S - K + 1, S - K + 1), device="cuda")
        s = torch.cuda.current_stream().cuda_stream
        xp, fp, yp = x.data_ptr(), f.data_ptr(), y.data_ptr()
        rows = []
        for v in (0, 1):
            _capi.debug_set_variant(v)
            rows.append((f"api v{v}", measure(lambda: pkg.conv2d_single(x, f, out=y))))
            rows.append((f"raw v{v}", measure(lambda: L.conv2d_single_ex(xp, S, S, fp, K, yp, s, 0))))
        _capi.debug_set_variant(0)
        rows.append(("torch y.add_", measure(lambda: y.add_(1.0))))
        print(f"{S}^2 K={K}: " + "  ".join(f"{n}: host {h:6.2f} dev {d:6.2f}" for n, (h, d) in rows), flush=True)


if __name__ == "__main__":
    main()

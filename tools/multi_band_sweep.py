#!/usr/bin/env python
"""conv2d_multi time per band height on the Table I layers and configs[2..3] (auto = the launch
heuristic). Prints ms per call for auto and for band counts 1, 2, 3, 4, 6, 8, 12, 16."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))
import torch  # noqa: E402

import paper_conf_cluster_luzw20_b200 as pkg  # noqa: E402
from gen import synth  # noqa: E402
from variants import time_call  # noqa: E402

TABLE1 = [("CONV1", 28, 128, 3), ("CONV2", 56, 64, 3), ("CONV3", 12, 64, 5), ("CONV4", 14, 16, 5),
          ("CONV5", 24, 256, 5), ("CONV6", 24, 64, 5), ("CONV7", 28, 16, 5), ("CONV8", 28, 512, 3),
          ("CONV9", 56, 256, 3), ("CONV10", 112, 128, 3), ("CONV11", 224, 64, 3)]


def main():
    layers = [(f"{nm} C{C}", 128, C, S, F, K) for C in (1, 3) for nm, S, F, K in TABLE1]
    layers += [("config2", 32, 64, 56, 64, 3), ("config3", 128, 3, 224, 64, 7)]
    for name, N, C, S, F, K in layers:
        x = synth.fill_torch(1, 1, (N, C, S, S), "img", device="cuda")
        w = torch.from_numpy(synth.make_filter(1, K, "he", F=F, C=C)).cuda()
        y = pkg.conv2d_multi(x, w)
        Ho = S - K + 1
        line = f"{name:12s} auto {time_call(lambda: pkg.conv2d_multi(x, w, out=y), 5) * 1e3:8.1f}"
        for b in (1, 2, 3, 4, 6, 8, 12, 16):
            if b > Ho:
                continue
            bh = -(-Ho // b)
            line += f"  b{b} {time_call(lambda: pkg.conv2d_multi(x, w, out=y, band_h=bh), 5) * 1e3:8.1f}"
        print(line, flush=True)


if __name__ == "__main__":
    main()

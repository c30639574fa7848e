"""One 8192^2 'same' call per K (for an ncu launch list of the padded path's kernels)."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_cluster_luzw20_b200 as pkg
from gen import synth
x = synth.fill_torch(1, 1, (8192, 8192), "img", device="cuda")
for K in (3, 5):
    f = torch.from_numpy(synth.make_filter(1, K, "rand")[0, 0]).cuda()
    for _ in range(2):
        pkg.conv2d_single_pad(x, f, "same_zero")
    torch.cuda.synchronize()

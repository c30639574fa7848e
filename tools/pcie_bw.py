#!/usr/bin/env python
"""Host<->device copy bandwidth (pinned), one direction and both at once: the e2e ceiling."""
import torch

n = 512 << 20  # bytes
h_in = torch.empty(n // 4, dtype=torch.float32).pin_memory()
h_out = torch.empty(n // 4, dtype=torch.float32).pin_memory()
d_a = torch.empty(n // 4, device="cuda")
d_b = torch.empty(n // 4, device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()


def timed(fn, reps=5):
    fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps


def both():
    s1.wait_stream(torch.cuda.current_stream())
    s2.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s1):
        d_a.copy_(h_in, non_blocking=True)
    with torch.cuda.stream(s2):
        h_out.copy_(d_b, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s1)
    torch.cuda.current_stream().wait_stream(s2)


t_h2d = timed(lambda: d_a.copy_(h_in, non_blocking=True))
t_d2h = timed(lambda: h_out.copy_(d_b, non_blocking=True))
t_both = timed(both)
print(f"H2D {n / t_h2d / 1e6:.1f} GB/s  D2H {n / t_d2h / 1e6:.1f} GB/s  both concurrently {2 * n / t_both / 1e6:.1f} GB/s total")

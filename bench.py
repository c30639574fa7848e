#!/usr/bin/env python
"""Benchmark of the hot path (driver contract).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference] [--workload NAME]
                    [--batch B]

Default workload = BASELINE.json configs[1], the workload its metric is quoted on: the single-channel
sweep of 1024^2, 2048^2, 4096^2, 8192^2 fp32 images x K in {3,5,7,9,11,13,15} (28 points). Each
point is a batch of B images (--batch, default 8) filtered with one filter: one conv2d_single_batch
call per point (conv2d_single when a rank holds one image), on its own input/output buffers, largest
images first. One "step" = one pass over all 28 points. `value` = output pixels of the whole job
/ time (Gpixel/s), timed on the device with CUDA events, max over ranks, L2 flushed (a 512 MiB write,
then a 256 MiB read that evicts its dirty lines) between steps outside the timed region.

Multi-GPU (--gpus N): one process per GPU over NCCL. Without torchrun's environment, bench.py
re-launches itself under `python -m torch.distributed.run --nproc-per-node N` (fails loudly when
fewer than N GPUs are visible). The batch of every point is split across ranks (shard.batch_range:
rank p takes images [p*B/N, (p+1)*B/N)) -- a fixed total amount of work, so "scaling": "strong", and
no data-path collective (north_star: "partitioned ... by image/batch ... no collective needed").
configs[2] / configs[3] (--workload config2 / config3) shard their N=32 / N=128 batches the same way;
configs[4] (--workload config4, one 32768^2 image, K=15) is split into row bands with the (K-1)-row
NCCL halo exchange of shard.py.

--impl reference: the CPU oracle (this tier's reference arm) timed as it stands on the host cores,
on a bounded sample of the same workload (rank 0 only).
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

BASELINE_METRIC = "conv2d Gpixel/s and multi-channel GFLOP/s (fp32) at 1/2/4/8 B200, % roofline"
SWEEP_SIZES = (8192, 4096, 2048, 1024)
SWEEP_KS = (3, 5, 7, 9, 11, 13, 15)
N_SM = 148
FMA_LANES_PER_SM = 128


def load_peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        with open(p) as fh:
            d = json.load(fh)
        return {"hbm_gbs": float(d["hbm_gbs"]), "sm_max_mhz": float(d.get("sm_max_mhz", 1965.0)),
                "bf16_tflops": float(d.get("bf16_tflops", 1590.0)),
                "source": "measured (MEASURED_PEAKS.json)"}
    except Exception:
        return {"hbm_gbs": 6650.0, "sm_max_mhz": 1965.0, "bf16_tflops": 1590.0,
                "source": "fallback (B200_PROFILING.md)"}


# nominal dense tf32 / bf16 tensor throughput ratio (B200_PROFILING.md: 1.1 vs 2.25 PFLOP/s)
TF32_PER_BF16 = 1.1 / 2.25


def fp32_fma_peak_tflops(sm_mhz):
    """fp32 CUDA-core peak: 148 SMs x 128 FMA lanes x 2 flop x clock."""
    return N_SM * FMA_LANES_PER_SM * 2 * sm_mhz * 1e6 / 1e12


# ------------------------------------------------------------------------------------------------
# workloads
# ------------------------------------------------------------------------------------------------
class Point:
    """One conv call of a step: shapes, device buffers, algorithmic work."""

    def __init__(self, kind, name, dims, K, padding="valid", flip=False, halo_rows=0, batch=1):
        self.kind, self.name, self.dims, self.K = kind, name, dims, K
        self.padding, self.flip, self.halo_rows = padding, flip, halo_rows  # N4 / N3 variants (single)
        self.batch = batch  # single: images per point (the whole job's batch); multi: dims[0]
        self.n0 = 0         # this rank's images [n0, n0 + n_local) of the batch (shard.batch_range)
        self.n_local = self.images
        self.x = self.f = self.y = self.halo = None

    @property
    def images(self):
        return self.batch if self.kind == "single" else self.dims[0]

    @property
    def out_px_image(self):
        """output elements of one image (single: pixels; multi: F output planes)"""
        if self.kind == "single":
            H, W = self.dims
            if self.padding != "valid":
                return H * W
            return (H - self.K + 1) * (W - self.K + 1)
        N, C, H, W, F = self.dims
        return F * (H - self.K + 1) * (W - self.K + 1)

    @property
    def out_px(self):
        """output elements of the whole point (all images of the batch)"""
        return self.out_px_image * self.images

    @property
    def flops(self):
        C = 1 if self.kind == "single" else self.dims[1]
        return 2.0 * self.out_px * C * self.K * self.K

    def local_units(self, unit):
        """units this rank computes per step"""
        per_img = self.out_px_image if unit == "Gpixel/s" else self.flops / self.images
        return per_img * self.n_local

    @property
    def bytes(self):
        """compulsory HBM bytes of the whole point: inputs + outputs + filters"""
        if self.kind == "single":
            H, W = self.dims
            return 4.0 * (self.batch * H * W + self.out_px + self.K * self.K)
        N, C, H, W, F = self.dims
        return 4.0 * (N * C * H * W + self.out_px + F * C * self.K * self.K)

    def in_bytes(self):
        """input bytes of this rank's images"""
        if self.kind == "single":
            return 4 * self.n_local * self.dims[0] * self.dims[1]
        N, C, H, W, F = self.dims
        return 4 * self.n_local * C * H * W

    def local_bound_seconds(self, peaks, sm_mhz):
        """roofline time of this rank's share of the point"""
        _, t = self.bound(peaks, sm_mhz)
        return t * self.n_local / max(1, self.images)

    def filt_bytes(self):
        C = 1 if self.kind == "single" else self.dims[1]
        F = 1 if self.kind == "single" else self.dims[4]
        return 4 * F * C * self.K * self.K

    def bound(self, peaks, sm_mhz):
        t_mem = self.bytes / (peaks["hbm_gbs"] * 1e9)
        t_fma = self.flops / (fp32_fma_peak_tflops(sm_mhz) * 1e12)
        return ("hbm", t_mem) if t_mem >= t_fma else ("alu", t_fma)


DEFAULT_SWEEP_BATCH = 8


def workload_points(name, batch=None):
    """The points of one step of a workload. batch: images per single-channel point (sweep default
    DEFAULT_SWEEP_BATCH, config0 default 1)."""
    if name == "sweep":
        b = DEFAULT_SWEEP_BATCH if batch is None else batch
        return [Point("single", f"{S}^2 K={K}", (S, S), K, batch=b) for S in SWEEP_SIZES for K in SWEEP_KS], \
            "Gpixel/s"
    if name == "config0":
        return [Point("single", "256^2 K=3", (256, 256), 3, batch=batch or 1)], "Gpixel/s"
    if name == "config2":
        return [Point("multi", "N32 C64 F64 56^2 K3", (32, 64, 56, 56, 64), 3)], "GFLOP/s"
    if name == "config3":
        return [Point("multi", "N128 C3 F64 224^2 K7", (128, 3, 224, 224, 64), 7)], "GFLOP/s"
    if name == "config4":
        return [Point("single", "32768^2 K=15", (32768, 32768), 15)], "Gpixel/s"
    if name == "pad":  # 'same' padding and true convolution
        return [Point("single", f"8192^2 K={K} {pad}{' flip' if flip else ''}", (8192, 8192), K, pad, flip)
                for K in (3, 15) for pad, flip in (("same_zero", False), ("same_replicate", True))], "Gpixel/s"
    if name == "halo":  # the last K-1 rows read in place from a separate allocation
        return [Point("single", f"8192^2 K={K} halo {K - 1} rows", (8192, 8192), K, halo_rows=K - 1)
                for K in (3, 15)], "Gpixel/s"
    if name == "table1":  # PAPER.md Table I: 11 layers x C in {1, 3}, N = 128
        return [Point("multi", f"{nm} C{C} N128 {S}^2 F{F} K{K}", (128, C, S, S, F), K)
                for C in (1, 3) for nm, S, F, K in TABLE1], "GFLOP/s"
    raise SystemExit(f"unknown workload {name}")


def shard_points(points, world, rank):
    """Split every point's batch across ranks (shard.batch_range): rank p computes images
    [n0, n0 + n_local). No data-path collective; the union over ranks is the whole job."""
    from paper_conf_cluster_luzw20_b200.shard import batch_range

    for p in points:
        n0, n1 = batch_range(p.images, world, rank)
        p.n0, p.n_local = n0, n1 - n0
    return points


def job_units(points, unit):
    """units of the whole job per step (all ranks)"""
    return sum(p.out_px if unit == "Gpixel/s" else p.flops for p in points)


# PAPER.md Table I: name, IH = IW, FN, FH = FW
TABLE1 = [("CONV1", 28, 128, 3), ("CONV2", 56, 64, 3), ("CONV3", 12, 64, 5), ("CONV4", 14, 16, 5),
          ("CONV5", 24, 256, 5), ("CONV6", 24, 64, 5), ("CONV7", 28, 16, 5), ("CONV8", 28, 512, 3),
          ("CONV9", 56, 256, 3), ("CONV10", 112, 128, 3), ("CONV11", 224, 64, 3)]

WORKLOAD_DESC = {
    "sweep": "BASELINE.json configs[1]: single-channel sweep, 1024^2/2048^2/4096^2/8192^2 x K in "
             "{3,5,7,9,11,13,15}, a batch of B images per point (28 conv2d_single_batch calls per step, "
             "largest first; the batch split across ranks)",
    "config0": "BASELINE.json configs[0]: 256x256, K=3 (batch B, default 1)",
    "config2": "BASELINE.json configs[2]: N=32, C=F=64, 56x56, K=3 (batch split across ranks)",
    "config3": "BASELINE.json configs[3]: N=128, C=3, F=64, 224x224, K=7 (batch split across ranks)",
    "config4": "BASELINE.json configs[4]: 32768x32768, K=15 (row bands + NCCL halo at N>1)",
    "table1": "PAPER.md Table I (P:335-352): 11 layers x C in {1,3}, N=128 (22 conv2d_multi calls per step)",
    "pad": "SURVEY 8(f) N4: 8192^2, K in {3,15}, 'same' zero padding / 'same' replicate padding + true "
           "convolution (conv2d_single_pad; 4 calls per step)",
    "halo": "SURVEY 8(f) N3: 8192^2, K in {3,15}, last K-1 rows in a separate allocation read in place "
            "(conv2d_single_halo, the fused row-band halo launch on one GPU; 2 calls per step)",
}


def materialise(points, device):
    """Device buffers of this rank's images of every point, generated in place from the global
    element index (gen/synth.py): the shards of all ranks together are the one-GPU batch, bit for bit."""
    import torch

    from gen import synth

    for i, p in enumerate(points):
        seed = synth.BASE_SEED + i
        if p.n_local == 0:
            continue
        if p.kind == "single":
            H, W = p.dims
            full = synth.fill_torch(seed, synth.TAG_INPUT, (p.n_local, H, W), "img", start=p.n0 * H * W,
                                    device=device)
            hr = p.halo_rows
            p.x = full[:, :H - hr].contiguous() if hr else full
            p.halo = full[:, H - hr:].contiguous() if hr else None
            del full
            p.f = torch.from_numpy(synth.make_filter(seed, p.K, "rand")[0, 0]).to(device)
            Ho, Wo = (H, W) if p.padding != "valid" else (H - p.K + 1, W - p.K + 1)
            p.y = torch.empty((p.n_local, Ho, Wo), device=device)
        else:
            N, C, H, W, F = p.dims
            p.x = synth.fill_torch(seed, synth.TAG_INPUT, (p.n_local, C, H, W), "img" if C < 8 else "sym",
                                   start=p.n0 * C * H * W, device=device)
            p.f = torch.from_numpy(synth.make_filter(seed, p.K, "he", F=F, C=C)).to(device)
            p.y = torch.empty((p.n_local, F, H - p.K + 1, W - p.K + 1), device=device)


# ------------------------------------------------------------------------------------------------
# clocks (NVML, sampled in a thread during the timed region)
# ------------------------------------------------------------------------------------------------
class ClockSampler:
    REASONS = {
        "gpu_idle": 0x1, "applications_clocks_setting": 0x2, "sw_power_cap": 0x4, "hw_slowdown": 0x8,
        "sync_boost": 0x10, "sw_thermal_slowdown": 0x20, "hw_thermal_slowdown": 0x40,
        "hw_power_brake_slowdown": 0x80, "display_clock_setting": 0x100,
    }

    def __init__(self, index, period_s=0.01):
        self.samples, self.reasons, self.max_mhz = [], set(), None
        self.period = period_s
        self._stop = threading.Event()
        self.ok = False
        try:
            import pynvml

            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(index)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
            self.ok = True
        except Exception as e:  # pragma: no cover
            self.err = str(e)

    def _run(self):
        while not self._stop.is_set():
            try:
                self.samples.append(self.nv.nvmlDeviceGetClockInfo(self.h, self.nv.NVML_CLOCK_SM))
                r = self.nv.nvmlDeviceGetCurrentClocksThrottleReasons(self.h)
                for k, bit in self.REASONS.items():
                    if r & bit and k != "gpu_idle":
                        self.reasons.add(k)
            except Exception:
                pass
            time.sleep(self.period)

    def __enter__(self):
        if self.ok:
            self.t = threading.Thread(target=self._run, daemon=True)
            self.t.start()
        return self

    def __exit__(self, *a):
        if self.ok:
            self._stop.set()
            self.t.join()

    def summary(self):
        if not self.ok or not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": self.max_mhz, "reasons": [], "samples": 0}
        return {"sm_mhz": statistics.median(self.samples), "sm_max_mhz": self.max_mhz,
                "reasons": sorted(self.reasons), "samples": len(self.samples)}


# ------------------------------------------------------------------------------------------------
# GPU arm
# ------------------------------------------------------------------------------------------------
def run_ours(args):
    import torch
    import torch.distributed as dist

    import paper_conf_cluster_luzw20_b200 as pkg
    from paper_conf_cluster_luzw20_b200 import shard

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if world != args.gpus:
        raise SystemExit(f"bench.py: --gpus {args.gpus} but WORLD_SIZE={world} (launch one rank per GPU)")
    if world > 1:
        if torch.cuda.device_count() < world:
            raise SystemExit(f"bench.py: {world} ranks but only {torch.cuda.device_count()} visible GPUs")
        torch.cuda.set_device(local)
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    device = torch.device("cuda", local)
    torch.cuda.set_device(device)
    peaks = load_peaks()

    points, unit = workload_points(args.workload, args.batch)
    if args.variant:
        pkg._capi.debug_set_variant(args.variant)  # tuning library (tools / A-B runs only)
    rowband = args.workload == "config4" and world > 1
    band = None
    if rowband:
        p = points[0]
        H, W = p.dims
        band = shard.row_band(H, W, p.K, world, rank)
        from gen import synth

        peer = None
        if args.halo == "p2p":  # band buffers in symmetric memory: the halo is read in place over NVLink
            p.x, peer, p2p_handle = shard.symmetric_band_buffers(band, device)
        elif args.halo == "ipc":  # same, buffers exchanged as CUDA IPC mappings (lazy peer access)
            p.x, peer, p2p_keep = shard.ipc_band_buffers(band, device)
        else:
            p.x = torch.empty((band.buf_rows, W), device=device)
        p.x[:band.in_rows] = synth.fill_torch(synth.BASE_SEED, synth.TAG_INPUT, (band.in_rows, W), "img",
                                              start=band.o0 * W, device=device)
        p.f = torch.from_numpy(synth.make_filter(synth.BASE_SEED, p.K, "gauss")[0, 0]).to(device)
        p.y = torch.empty((band.out_rows, W - p.K + 1), device=device)
        p.n0, p.n_local = 0, 1
        if args.halo in ("p2p", "ipc"):  # every neighbour's rows are written before any rank reads them
            torch.cuda.synchronize()
            dist.barrier()
    else:
        shard_points(points, world, rank)
        materialise(points, device)
    stream = torch.cuda.current_stream(device)
    flush = torch.empty(512 * (1 << 20) // 4, dtype=torch.float32, device=device)
    flush_rd = torch.ones(256 * (1 << 20) // 4, dtype=torch.float32, device=device)

    def l2_flush():
        # write 512 MiB (> 126 MB L2), then read 256 MiB: the read evicts the dirty lines of the write,
        # so their write-back happens here and not inside the next timed kernel
        flush.zero_()
        flush_rd.max()

    use_graph = not rowband and (args.graph == "on" or (args.graph == "auto" and args.workload == "config0"))
    capturing = [False]
    active = [i for i, p in enumerate(points) if p.n_local > 0]

    def run_point(p, on=None):
        st = None if capturing[0] else (on if on is not None else stream)  # capture: torch's capture stream
        if rowband and args.halo in ("p2p", "ipc"):
            shard.rowband_conv2d_single_p2p(p.x, peer, p.f, band, p.y)
        elif rowband:
            shard.rowband_conv2d_single(p.x, p.f, band, p.y)
        elif p.kind == "single" and p.halo is not None:
            pkg.conv2d_single_halo(p.x[0], p.halo[0], p.f, out=p.y[0], stream=st)
        elif p.kind == "single" and (p.padding != "valid" or p.flip):
            pkg.conv2d_single_pad(p.x[0], p.f, p.padding, p.flip, out=p.y[0], stream=st)
        elif p.kind == "single" and p.n_local == 1:
            pkg.conv2d_single(p.x[0], p.f, out=p.y[0], stream=st)
        elif p.kind == "single":
            pkg.conv2d_single_batch(p.x, p.f, out=p.y, stream=st)
        elif args.multi_impl == "tc":
            pkg.conv2d_multi_tc(p.x, p.f, out=p.y, stream=st)
        else:
            pkg.conv2d_multi(p.x, p.f, out=p.y, stream=st)

    n = len(points)

    # Concurrency of the timed steps (--concurrency small): the largest convolutions (the 8192^2 points
    # of the sweep, incl. the dominant kernel) run one after the other on the main stream, so each fills
    # the GPU alone and the dominant kernel's events time it in isolation; the smaller, latency-bound
    # ones -- independent images -- are then spread over one stream per K (each K has its own
    # constant-memory filter slot, so no two streams contend for one) and joined back.
    def in_px(p):
        return p.dims[0] * p.dims[1] if p.kind == "single" else p.dims[0] * p.dims[2] * p.dims[3]

    px_max = max(in_px(points[i]) for i in active) if active else 0
    lanes = {}
    conc = args.concurrency if args.concurrency != "auto" else ("small" if args.workload == "table1" else "serial")
    if conc == "small" and not rowband and not use_graph:
        for i in active:
            if in_px(points[i]) < px_max:
                lanes.setdefault(points[i].K, torch.cuda.Stream(device))

    def step(evs=None, dom=None, dom_evs=None):
        """one pass over the workload; evs: an event after every point (warm-up breakdown);
        dom/dom_evs: events bracketing the dominant point only (timed steps: 2 extra events)"""
        if lanes and evs is None:
            big = [i for i in active if in_px(points[i]) == px_max]
            small = [i for i in active if in_px(points[i]) < px_max]
            for i in big:
                if dom_evs is not None and i == dom:
                    dom_evs[0].record(stream)
                run_point(points[i])
                if dom_evs is not None and i == dom:
                    dom_evs[1].record(stream)
            fork = torch.cuda.Event()
            fork.record(stream)
            for ln in lanes.values():
                ln.wait_event(fork)
            for i in small:
                ln = lanes[points[i].K]
                if dom_evs is not None and i == dom:
                    dom_evs[0].record(ln)
                run_point(points[i], ln)
                if dom_evs is not None and i == dom:
                    dom_evs[1].record(ln)
            for ln in lanes.values():
                j = torch.cuda.Event()
                j.record(ln)
                stream.wait_event(j)
            return
        for i in range(n):
            if dom_evs is not None and i == dom:
                dom_evs[0].record(stream)
            if i in active_set:
                run_point(points[i])
            if dom_evs is not None and i == dom:
                dom_evs[1].record(stream)
            if evs is not None:
                evs[i + 1].record(stream)

    active_set = set(active)
    # warm-up steps: per-point events give the per-point breakdown and pick the dominant kernel
    warm_ms = [0.0] * n
    counted = max(1, args.warmup - 1)  # the first warm-up step pays one-time setup: not counted
    for w in range(args.warmup):
        l2_flush()
        evs = [torch.cuda.Event(enable_timing=True) for _ in range(n + 1)]
        evs[0].record(stream)
        step(evs)
        torch.cuda.synchronize()
        if w > 0 or args.warmup == 1:
            for i in range(n):
                warm_ms[i] += evs[i].elapsed_time(evs[i + 1]) / counted
    dom = max(range(n), key=lambda i: warm_ms[i] if i in active_set else -1.0)
    if lanes:  # one untimed step in the timed steps' (concurrent) form
        l2_flush()
        step()
    torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()

    graph = None
    if use_graph:
        # latency-bound workload (one small image): the step is captured once into a CUDA graph and
        # replayed, so the timed region holds the device work, not the Python/driver call overhead
        graph = torch.cuda.CUDAGraph()
        capturing[0] = True
        with torch.cuda.graph(graph):
            step()
        capturing[0] = False
        graph.replay()
        torch.cuda.synchronize()

    # timed steps: barrier + synchronize on both sides; events at the step boundaries and around the
    # dominant kernel only
    step_events = [[torch.cuda.Event(enable_timing=True) for _ in range(4)] for _ in range(args.steps)]
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    with ClockSampler(local) as clk:
        for s in range(args.steps):
            l2_flush()  # L2 flush, outside [ev0, ev3]
            ev = step_events[s]
            ev[0].record(stream)
            if graph is not None:  # one point per step: the dominant kernel is the whole replay
                ev[1].record(stream)
                graph.replay()
                ev[2].record(stream)
            else:
                step(dom=dom, dom_evs=(ev[1], ev[2]))
            ev[3].record(stream)
        torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()

    total_ms = sum(ev[0].elapsed_time(ev[3]) for ev in step_events)
    dom_ms = sum(ev[1].elapsed_time(ev[2]) for ev in step_events) / args.steps
    per_point_ms = list(warm_ms)
    launches_local = sum(1 for _ in active) * args.steps * (2 if rowband and args.halo == "nccl" and not band.is_last
                                                            else 1)
    if world > 1:  # max over ranks of the timed region; sum of the kernel launches
        t = torch.tensor([total_ms], dtype=torch.float64, device=device)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        total_ms = float(t.item())
        c = torch.tensor([launches_local], dtype=torch.int64, device=device)
        dist.all_reduce(c, op=dist.ReduceOp.SUM)
        launches = int(c.item())
    else:
        launches = launches_local

    units_per_step = job_units(points, unit)  # the whole job: every rank's share (row bands: the one image)
    value = units_per_step * args.steps / (total_ms * 1e-3) / 1e9

    clocks = clk.summary()
    sm_mhz_peak = peaks["sm_max_mhz"]

    # roofline of the dominant kernel (largest share of this rank's step), timed inside the timed steps:
    # this rank's share of the point (its images, or its row band)
    dp = points[dom]
    dkind, _ = dp.bound(peaks, sm_mhz_peak)
    dsec = dom_ms * 1e-3
    share = (band.out_rows / (dp.dims[0] - dp.K + 1)) if rowband else dp.n_local / max(1, dp.images)
    d_flops, d_bytes = dp.flops * share, dp.bytes * share
    if dp.kind == "multi" and args.multi_impl == "tc":
        # tensor-core variant: the executed TF32 MMA flops (3 per useful product, the 3xTF32 split)
        # against the tf32 tensor peak (measured bf16 burst x the nominal tf32/bf16 ratio)
        roof = {"bound": "tensor", "achieved": 3 * d_flops / dsec / 1e12,
                "peak": peaks["bf16_tflops"] * TF32_PER_BF16, "unit": "TFLOP/s",
                "note": "executed tf32 MMA TFLOP/s = 3 x useful (3xTF32); peak = bf16 burst x 1.1/2.25"}
    elif dkind == "hbm":
        roof = {"bound": "hbm", "achieved": d_bytes / dsec / 1e9, "peak": peaks["hbm_gbs"], "unit": "GB/s"}
    else:
        roof = {"bound": "alu", "achieved": d_flops / dsec / 1e12, "peak": fp32_fma_peak_tflops(sm_mhz_peak),
                "unit": "TFLOP/s"}
    roof["frac"] = roof["achieved"] / roof["peak"]
    roof["kernel"] = (f"conv2d_multi_tc {dp.name}" if dp.kind == "multi" and args.multi_impl == "tc"
                      else f"conv2d_{dp.kind} {dp.name}" + (f" x{dp.n_local} images" if dp.kind == "single"
                                                            and dp.n_local > 1 else ""))
    roof["share_of_step"] = dom_ms / max(total_ms / args.steps, 1e-12)
    roof["launch_ms"] = round(dom_ms, 5)
    roof["peak_source"] = (peaks["source"] if dkind == "hbm" or roof["bound"] == "tensor" else
                           f"fp32 FMA: 148 SM x 128 lanes x 2 x {sm_mhz_peak:.0f} MHz (sm_max_mhz, "
                           f"{peaks['source']})")
    roof["traffic"] = load_traffic(roof["kernel"])

    sweep = []
    for i, p in enumerate(points):
        if i not in active_set:
            continue
        kind, _ = p.bound(peaks, sm_mhz_peak)
        t = per_point_ms[i] * 1e-3
        t_roof = (p.local_bound_seconds(peaks, sm_mhz_peak) if not rowband else
                  p.bound(peaks, sm_mhz_peak)[1] * share)
        u = (p.local_units(unit) if not rowband else p.out_px * share)
        sweep.append({"point": p.name, "images": p.n_local, "ms": round(per_point_ms[i], 5),
                      ("gpx_s" if unit == "Gpixel/s" else "gflop_s"): round(u / t / 1e9, 2),
                      "bound": kind, "roofline_frac": round(t_roof / t, 4)})
    t_roof_step = sum(points[i].local_bound_seconds(peaks, sm_mhz_peak) for i in active) if not rowband else None

    batched = points[0].kind == "single" and not rowband and args.workload in ("sweep", "config0")
    line = {
        "metric": BASELINE_METRIC,
        "metric_detail": f"{unit} of the {args.workload} workload (whole job, all ranks)",
        "value": round(value, 3),
        "unit": unit,
        "n_gpus": world,
        "steps": args.steps,
        "warmup": args.warmup,
        "ms_per_step": round(total_ms / args.steps, 5),
        "higher_is_better": True,
        "scaling": "strong" if (world > 1 or rowband or args.workload in ("sweep", "config2", "config3", "config0"))
        else "weak",
        "vs_baseline": None,
        "dtype": "f32",
        "data": "synthetic (seeded counter-based generator, gen/synth.py)",
        "config": {"workload": WORKLOAD_DESC[args.workload],
                   **({"batch": points[0].batch} if batched else {}),
                   **({"multi_impl": args.multi_impl} if points[0].kind == "multi" else {}),
                   "l2": "512 MiB write + 256 MiB read between timed steps (outside the events) + distinct buffers per "
                         "point; 8192^2 inputs also exceed L2",
                   "parallelism": (("row bands + NCCL halo" if args.halo == "nccl" else
                                    f"row bands, halo read in place from the neighbour ({args.halo}, NVLink)")
                                   if rowband else
                                   (f"batch split over {world} ranks (shard.batch_range), no collective"
                                    if world > 1 else "1 GPU")),
                   "filter": "rand (2u-1)/K" if points[0].kind == "single" else "he",
                   "input": "img u in [0,1)"},
        "roofline": roof,
        "roofline_step_frac": (round(t_roof_step / (total_ms / args.steps * 1e-3), 4) if t_roof_step else None),
        "gpu_launches": launches,
        "clocks": clocks,
        "points_warmup": sweep,
        "points_note": "per-point times (this rank) from the warm-up steps (an event after every call); the timed "
                       "steps carry events only at the step boundaries and around the dominant kernel",
    }
    if lanes:
        line["config"]["concurrency"] = (f"the {sum(in_px(points[i]) == px_max for i in active)} largest calls "
                                         f"serially on one stream, the others on {len(lanes)} streams (one per K), "
                                         f"joined every step")
    if graph is not None:
        line["config"]["timing"] = ("CUDA graph of the step (captured once, replayed per timed step): "
                                    "device time without per-call host overhead")

    # end to end through the public API with host buffers (pinned), copies inside the timed region
    if not rowband and not args.no_e2e:
        e2e = run_e2e([points[i] for i in active], unit, args, device)
        if world > 1:  # whole job: every rank moved its own images; time = max over ranks
            t = torch.tensor([e2e["ms_per_step"], e2e["h2d_bytes_per_step"], e2e["d2h_bytes_per_step"]],
                             dtype=torch.float64, device=device)
            tm = t[:1].clone()
            dist.all_reduce(tm, op=dist.ReduceOp.MAX)
            tb = t[1:].clone()
            dist.all_reduce(tb, op=dist.ReduceOp.SUM)
            ms = float(tm.item())
            e2e["value"] = round(units_per_step * e2e["steps"] / (ms * e2e["steps"] * 1e-3) / 1e9, 3)
            e2e["ms_per_step"] = round(ms, 3)
            e2e["h2d_bytes_per_step"] = int(tb[0].item())
            e2e["d2h_bytes_per_step"] = int(tb[1].item())
        line["e2e"] = e2e

    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        line["cpu_baseline"] = cpu_baseline(args.workload, budget_s=args.cpu_budget, batch=args.batch)

    if world > 1:
        dist.barrier()
        dist.destroy_process_group()
    if rank == 0:
        print(json.dumps(line), flush=True)


def run_e2e(points, unit, args, device):
    """Same metric through the user-facing host-buffer call (C ABI conv2d_single_host: chunked
    H2D / kernel / D2H pipeline, one call per image; multi-channel: torch copies around conv2d_multi),
    pinned host tensors, every byte of every input copied in and every output copied out inside the
    events. Consecutive calls alternate between two streams (independent images), as a user pipelining
    a batch of images would, so one call's device->host copies overlap the next call's host->device."""
    # Keep the host side on the GPU's NUMA node: the pinned staging buffers are first-touched by
    # this thread, so they land in memory local to the GPU's PCIe root (cross-socket DMA halves the
    # copy bandwidth and made the number swing run to run). Restored afterwards.
    old_aff = os.sched_getaffinity(0)
    try:
        import pynvml

        pynvml.nvmlInit()
        h = pynvml.nvmlDeviceGetHandleByIndex(device.index or 0)
        words = pynvml.nvmlDeviceGetCpuAffinity(h, (os.cpu_count() + 63) // 64)
        local = {w * 64 + b for w, m in enumerate(words) for b in range(64) if m >> b & 1}
        local &= old_aff
        if local:
            os.sched_setaffinity(0, local)
    except Exception:
        pass
    try:
        return _run_e2e(points, unit, args, device)
    finally:
        os.sched_setaffinity(0, old_aff)


def _run_e2e(points, unit, args, device):
    import torch

    import paper_conf_cluster_luzw20_b200 as pkg

    main = torch.cuda.current_stream(device)
    ns = max(1, args.e2e_streams)
    streams = [torch.cuda.Stream(device=device) for _ in range(ns)]
    # host buffers: one pinned input / output per distinct shape (the host side has no L2 to defeat)
    hx, hy = {}, {}
    for p in points:
        key = (p.kind, p.dims, p.K)
        if p.kind == "single" and (p.dims, p.n_local) not in hx:
            hx[(p.dims, p.n_local)] = p.x.cpu().pin_memory()
        elif p.kind == "multi":
            hx[key] = p.x.cpu().pin_memory()
        hy[key] = torch.empty(tuple(p.y.shape), dtype=torch.float32, pin_memory=True)
    hf = [p.f.cpu().pin_memory() for p in points]
    steps = max(1, min(args.steps, args.e2e_steps))

    def one():
        for s in streams:
            s.wait_stream(main)
        c = 0
        for i, p in enumerate(points):
            key = (p.kind, p.dims, p.K)
            if p.kind == "single":
                xin, yout = hx[(p.dims, p.n_local)], hy[key]
                for j in range(p.n_local):
                    pkg.conv2d_single_host(xin[j], hf[i], device=device, stream=streams[c % ns], out_host=yout[j])
                    c += 1
            else:
                pkg.conv2d_multi_host(hx[key], hf[i], device=device, stream=streams[c % ns], out_host=hy[key],
                                      impl=args.multi_impl)
                c += 1
        for s in streams:
            main.wait_stream(s)

    for _ in range(2):  # warm-up: pinned-page first touch, allocator pool growth
        one()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(main)
    for _ in range(steps):
        one()
    e1.record(main)
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1)
    units = sum(p.local_units(unit) for p in points) * steps
    h2d = sum(p.in_bytes() + p.filt_bytes() * (p.n_local if p.kind == "single" else 1) for p in points)
    d2h = sum(4 * p.y.numel() for p in points)
    return {"value": round(units / (ms * 1e-3) / 1e9, 3), "unit": unit, "h2d_bytes_per_step": h2d,
            "d2h_bytes_per_step": d2h, "steps": steps, "ms_per_step": round(ms / steps, 3),
            "path": (f"conv2d_single_host (C ABI, pinned host buffers, one call per image, {ns} streams)"
                     if points[0].kind == "single" else
                     f"conv2d_multi_host (impl={args.multi_impl}; pinned host buffers, {ns} streams)")}


def load_traffic(kernel_name):
    """dram bytes (read + write) per launch of this kernel config (bench roofline "kernel" name) from the
    committed ncu capture (profiles/ncu_traffic.json, tools/make_profiles.py)."""
    path = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    try:
        with open(path) as fh:
            d = json.load(fh)
        return d.get(kernel_name)
    except Exception:
        return None


# ------------------------------------------------------------------------------------------------
# CPU oracle legs (cpu_baseline and --impl reference) -- the only bench code touching oracle/
# ------------------------------------------------------------------------------------------------
def _oracle_sample(points, frac):
    """Run the oracle on the first ceil(frac * rows) output rows (single) / images (multi) of every
    point; inputs for just those rows are generated on the host. Returns (units, seconds)."""
    import numpy as np

    import oracle
    from gen import synth

    units = 0.0
    secs = 0.0
    for i, p in enumerate(points):
        seed = synth.BASE_SEED + i
        if p.kind == "single":
            H, W = p.dims
            Ho = H - p.K + 1
            rows = max(1, math.ceil(frac * Ho))
            x = synth.fill_np(seed, synth.TAG_INPUT, (rows + p.K - 1, W), "img")
            f = synth.make_filter(seed, p.K, "rand")[0, 0]
            t0 = time.perf_counter()
            if p.padding != "valid" or p.flip:
                y, _, _ = oracle.conv2d_single_pad(x, f, p.padding, p.flip)
            else:
                y, _, _ = oracle.conv2d_single(x, f, want_bound=False)
            secs += time.perf_counter() - t0
            units += y.size
        else:
            N, C, H, W, F = p.dims
            imgs = max(1, math.ceil(frac * N))
            x = synth.fill_np(seed, synth.TAG_INPUT, (imgs, C, H, W), "img" if C < 8 else "sym")
            w = synth.make_filter(seed, p.K, "he", F=F, C=C)
            t0 = time.perf_counter()
            oracle.conv2d_multi(x, w, want_bound=False)
            secs += time.perf_counter() - t0
            units += 2.0 * imgs * F * (H - p.K + 1) * (W - p.K + 1) * C * p.K * p.K
    return units, secs


def _set_omp():
    os.environ.setdefault("OMP_NUM_THREADS", str(len(os.sched_getaffinity(0))))


def _calibrate(points, budget_s):
    """Pick the sample fraction so the oracle sample takes about budget_s seconds (capped at 1)."""
    total_rows = sum((p.dims[0] - p.K + 1) if p.kind == "single" else p.dims[0] for p in points)
    frac = min(1.0, 2.0 * len(points) / total_rows)  # a couple of rows per point
    u, s = _oracle_sample(points, frac)
    while s < 0.5 and frac < 1.0:
        frac = min(1.0, frac * 4)
        u, s = _oracle_sample(points, frac)
    return min(1.0, frac * budget_s / max(s, 1e-6)), u, s


def cpu_baseline(workload, budget_s=10.0, batch=None):
    _set_omp()
    import oracle

    points, unit = workload_points(workload, batch)
    frac, _, _ = _calibrate(points, budget_s)
    u, s = _oracle_sample(points, frac)
    what = "output rows of the first image" if points[0].kind == "single" else "images"
    return {"value": round(u / s / 1e9, 6), "unit": unit, "cores": oracle.num_threads(), "kind": "oracle",
            "sample": f"first {frac * 100:.3g}% of the {what} of every point of the {workload} workload "
                      f"({s:.1f} s of oracle time; double accumulation, OpenMP over output rows)",
            "seconds": round(s, 2)}


def run_reference(args):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return  # under torchrun only rank 0 runs the CPU reference
    _set_omp()
    import oracle

    points, unit = workload_points(args.workload, args.batch)
    budget = max(0.5, args.ref_budget / max(1, args.steps + args.warmup))
    frac, _, _ = _calibrate(points, budget)
    for _ in range(args.warmup):
        _oracle_sample(points, frac)
    tot_u = tot_s = 0.0
    for _ in range(args.steps):
        u, s = _oracle_sample(points, frac)
        tot_u += u
        tot_s += s
    value = tot_u / tot_s / 1e9
    what = "output rows of the first image" if points[0].kind == "single" else "images"
    sample = (f"each step: first {frac * 100:.3g}% of the {what} of every point of the {args.workload} "
              f"workload (bounded sample; the full step would take ~{tot_s / args.steps / frac:.0f} s)")
    print(json.dumps({
        "impl": "reference",
        "metric": BASELINE_METRIC,
        "metric_detail": f"{unit} of the {args.workload} workload, CPU oracle",
        "value": round(value, 6), "unit": unit, "n_gpus": int(os.environ.get("WORLD_SIZE", "1")),
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": round(tot_s / args.steps * 1e3, 3),
        "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "f64",
        "data": "synthetic (seeded counter-based generator, gen/synth.py)",
        "config": {"workload": WORKLOAD_DESC[args.workload], "sample_fraction": frac},
        "cpu_baseline": {"value": round(value, 6), "unit": unit, "cores": oracle.num_threads(),
                         "kind": "oracle", "sample": sample},
        "e2e": {"value": round(value, 6), "unit": unit, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
        "gpu_launches": 0,
    }), flush=True)


def torchrun_cmd(argv, gpus, port):
    """The command that re-launches this script with one process per GPU (the driver's own form)."""
    return [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={gpus}",
            "--master-addr", "127.0.0.1", f"--master-port={port}", os.path.abspath(__file__), *argv]


def _free_port():
    import socket

    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--workload", default="sweep", choices=sorted(WORKLOAD_DESC))
    ap.add_argument("--batch", type=int, default=None,
                    help=f"images per single-channel point (sweep default {DEFAULT_SWEEP_BATCH}, config0 default 1); "
                         "split across ranks")
    ap.add_argument("--e2e-steps", type=int, default=3)
    ap.add_argument("--e2e-streams", type=int, default=2, help="e2e: caller streams the per-image host calls alternate over")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--cpu-budget", type=float, default=10.0)
    ap.add_argument("--ref-budget", type=float, default=90.0)
    ap.add_argument("--variant", type=int, default=0, help="tuning: force a single-channel kernel variant")
    ap.add_argument("--halo", choices=["nccl", "p2p", "ipc"], default="nccl",
                    help="config4 at N>1: NCCL P2P halo exchange (+ tail call), or the fused in-place halo read "
                         "from the neighbour's band mapped by symmetric memory (p2p) or CUDA IPC (ipc)")
    ap.add_argument("--concurrency", choices=["auto", "small", "serial"], default="auto",
                    help="timed steps: the largest convolutions serially, the smaller independent ones on one "
                         "stream per K (small), or every call in order on one stream (serial); auto: small for "
                         "table1 (measured +6%%), serial elsewhere (the sweep measured neutral)")
    ap.add_argument("--graph", choices=["auto", "on", "off"], default="auto",
                    help="replay the step as a CUDA graph (auto: config0, the latency-bound single 256^2 call)")
    ap.add_argument("--multi-impl", choices=["cuda", "tc"], default="cuda",
                    help="multi-channel workloads: conv2d_multi (CUDA cores) or conv2d_multi_tc (tcgen05 3xTF32)")
    args = ap.parse_args()
    if args.warmup < 3 and args.impl == "ours":
        args.warmup = 3  # contract: W >= 3
    if args.batch is not None and args.batch < 1:
        raise SystemExit("--batch must be >= 1")
    if args.workload in ("pad", "halo"):
        args.no_e2e = True  # the host-buffer entry (e2e) is the valid-mode one-segment call
    if args.impl == "reference":
        run_reference(args)
        return
    if args.gpus > 1 and "WORLD_SIZE" not in os.environ:
        # one process per GPU: re-launch under torchrun (the driver launches us that way itself)
        import torch

        have = torch.cuda.device_count()
        if have < args.gpus:
            raise SystemExit(f"bench.py: --gpus {args.gpus} needs {args.gpus} visible GPUs, found {have}")
        cmd = torchrun_cmd(sys.argv[1:], args.gpus, _free_port())
        os.execvp(cmd[0], cmd)
    run_ours(args)


if __name__ == "__main__":
    main()

"""Host-side checks of bench.py's workload definitions (no GPU): every workload resolves, the units
per step and the compulsory bytes follow SURVEY 8(d), and the N3 / N4 workloads count their outputs
correctly ('same' output = H x W)."""
import importlib.util
import os

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def bench():
    spec = importlib.util.spec_from_file_location("bench", os.path.join(ROOT, "bench.py"))
    mod = importlib.util.module_from_spec(spec)
    spec.loader.exec_module(mod)
    return mod


def test_every_workload_resolves(bench):
    for name in bench.WORKLOAD_DESC:
        points, unit = bench.workload_points(name)
        assert points and unit in ("Gpixel/s", "GFLOP/s")


def test_sweep_is_configs1(bench):
    points, unit = bench.workload_points("sweep")
    assert unit == "Gpixel/s" and len(points) == 28
    assert {p.dims for p in points} == {(s, s) for s in (1024, 2048, 4096, 8192)}
    assert {p.K for p in points} == {3, 5, 7, 9, 11, 13, 15}


def test_units_and_bytes(bench):
    p = bench.Point("single", "x", (100, 50), 5)
    assert p.out_px == 96 * 46 and p.flops == 2.0 * 96 * 46 * 25
    assert p.bytes == 4.0 * (100 * 50 + 96 * 46 + 25)
    q = bench.Point("single", "x", (100, 50), 5, padding="same_zero")
    assert q.out_px == 100 * 50
    m = bench.Point("multi", "x", (2, 3, 20, 30, 4), 3)
    assert m.out_px == 2 * 4 * 18 * 28 and m.flops == 2.0 * m.out_px * 3 * 9
    pad, _ = bench.workload_points("pad")
    assert all(p.padding != "valid" for p in pad)
    halo, _ = bench.workload_points("halo")
    assert all(p.halo_rows == p.K - 1 for p in halo)


def test_sweep_batch_and_sharding(bench):
    """The sweep's batch is split across ranks with no overlap and no gap; the whole-job units do
    not depend on the rank count (strong scaling: the driver's per-N values are comparable)."""
    points, unit = bench.workload_points("sweep")
    assert all(p.batch == bench.DEFAULT_SWEEP_BATCH for p in points)
    total = bench.job_units(points, unit)
    assert total == sum((p.dims[0] - p.K + 1) * (p.dims[1] - p.K + 1) * p.batch for p in points)
    for world in (1, 2, 3, 4, 8, 16):
        covered = {}
        local_sum = 0
        for rank in range(world):
            pts, _ = bench.workload_points("sweep")
            bench.shard_points(pts, world, rank)
            local_sum += sum(p.local_units(unit) for p in pts)
            for i, p in enumerate(pts):
                for n in range(p.n0, p.n0 + p.n_local):
                    assert (i, n) not in covered
                    covered[(i, n)] = rank
        assert len(covered) == len(points) * bench.DEFAULT_SWEEP_BATCH
        assert local_sum == total
    c3, u3 = bench.workload_points("config3")
    bench.shard_points(c3, 8, 7)
    assert c3[0].n_local == 16 and c3[0].n0 == 112
    assert abs(c3[0].local_units(u3) * 8 - bench.job_units(c3, u3)) < 1e-3 * bench.job_units(c3, u3)


def test_torchrun_relaunch_command(bench):
    cmd = bench.torchrun_cmd(["--gpus", "4", "--steps", "5"], 4, 29512)
    assert cmd[1:4] == ["-m", "torch.distributed.run", "--nnodes=1"]
    assert "--nproc-per-node=4" in cmd and "127.0.0.1" in cmd and "--master-port=29512" in cmd
    assert cmd[-4:] == ["--gpus", "4", "--steps", "5"] and cmd[-5].endswith("bench.py")


def _rank_units(rank, world, port, out):
    import importlib.util

    import torch
    import torch.distributed as dist

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        spec = importlib.util.spec_from_file_location("bench", os.path.join(ROOT, "bench.py"))
        b = importlib.util.module_from_spec(spec)
        spec.loader.exec_module(b)
        for wl in ("sweep", "config2", "config3"):
            pts, unit = b.workload_points(wl)
            b.shard_points(pts, world, rank)
            t = torch.tensor([sum(p.local_units(unit) for p in pts)], dtype=torch.float64)
            dist.all_reduce(t)  # the bench sums nothing on the data path; this checks the accounting
            if rank == 0:
                out[wl] = (float(t.item()), float(b.job_units(pts, unit)))
    finally:
        dist.destroy_process_group()


def test_rank_accounting_gloo():
    """world_size 2 and 3 over gloo: the units the ranks compute add up to the whole job."""
    import socket

    import torch.multiprocessing as mp

    for world in (2, 3):
        with socket.socket() as s:
            s.bind(("127.0.0.1", 0))
            port = s.getsockname()[1]
        mgr = mp.Manager()
        out = mgr.dict()
        mp.spawn(_rank_units, args=(world, port, out), nprocs=world, join=True)
        for wl, (summed, total) in out.items():
            assert abs(summed - total) <= 1e-9 * total, (world, wl)
        assert set(out.keys()) == {"sweep", "config2", "config3"}

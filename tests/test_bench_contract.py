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

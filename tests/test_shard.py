"""Host-side multi-GPU logic on CPU: partition arithmetic, and the row-band halo exchange and batch /
filter sharding run as world_size 2 and 3 process groups over gloo. The compute callback is the CPU
oracle here (tests may call it; the product default is the CUDA C-ABI call). Sharded results must be
bitwise equal to the unsharded oracle result."""
import os
import socket
import tempfile

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from gen import synth
from paper_conf_cluster_luzw20_b200 import shard


def test_even_split():
    for n in (0, 1, 7, 64, 1000):
        for world in (1, 2, 3, 8):
            parts = [shard.even_split(n, world, r) for r in range(world)]
            assert parts[0][0] == 0 and parts[-1][1] == n
            assert all(parts[i][1] == parts[i + 1][0] for i in range(world - 1))
            sizes = [b - a for a, b in parts]
            assert max(sizes) - min(sizes) <= 1


def test_row_band_geometry():
    H, W, K = 32768, 32768, 15
    bands = [shard.row_band(H, W, K, 8, r) for r in range(8)]
    assert bands[0].o0 == 0 and bands[-1].o1 == H - K + 1
    assert sum(b.in_rows for b in bands) == H  # every input row generated exactly once
    for b in bands:
        assert b.buf_rows == b.out_rows + K - 1
    with pytest.raises(ValueError):
        shard.row_band(20, 20, 15, 4, 0)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _oracle_compute(x, f, out):
    import oracle

    y, _, _ = oracle.conv2d_single(x.numpy(), f.numpy())
    out.copy_(torch.from_numpy(y))


def _worker_rowband(rank, world, port, H, W, K, tmpdir):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        band = shard.row_band(H, W, K, world, rank)
        buf = torch.full((band.buf_rows, W), float("nan"))
        # each rank generates only its own input rows, from the global-index generator
        buf[:band.in_rows] = torch.from_numpy(
            synth.fill_np(11, synth.TAG_INPUT, (band.in_rows, W), "img", start=band.o0 * W))
        f = torch.from_numpy(synth.make_filter(11, K, "rand")[0, 0])
        out = torch.empty((band.out_rows, W - K + 1))
        shard.rowband_conv2d_single(buf, f, band, out, compute=_oracle_compute)
        np.save(os.path.join(tmpdir, f"band{rank}.npy"), out.numpy())
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,K", [(2, 5), (3, 15), (2, 1)])
def test_rowband_halo_exchange_gloo(world, K):
    import oracle

    H, W = 64, 37
    with tempfile.TemporaryDirectory() as tmp:
        mp.spawn(_worker_rowband, args=(world, _free_port(), H, W, K, tmp), nprocs=world, join=True)
        got = np.concatenate([np.load(os.path.join(tmp, f"band{r}.npy")) for r in range(world)])
    x = synth.fill_np(11, synth.TAG_INPUT, (H, W), "img")
    ref, _, _ = oracle.conv2d_single(x, synth.make_filter(11, K, "rand")[0, 0])
    assert np.array_equal(got, ref)


def _oracle_compute_halo(x, halo, f, out):
    _oracle_compute(torch.cat([x, halo]), f, out)


def _worker_rowband_p2p(rank, world, port, H, W, K, tmpdir):
    """The fused-halo path: each rank reads rank+1's first K-1 rows where they are. On CPU the
    peer-memory view is stood in for by a separate tensor filled over gloo (symmetric memory needs
    GPUs); the compute call gets own rows and halo as two separate segments."""
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        band = shard.row_band(H, W, K, world, rank)
        buf = torch.from_numpy(synth.fill_np(11, synth.TAG_INPUT, (band.in_rows, W), "img", start=band.o0 * W))
        f = torch.from_numpy(synth.make_filter(11, K, "rand")[0, 0])
        peer = torch.full((band.halo, W), float("nan"))
        ops = []
        if rank > 0 and band.halo:
            ops.append(dist.P2POp(dist.isend, buf[:band.halo].contiguous(), rank - 1))
        if not band.is_last and band.halo:
            ops.append(dist.P2POp(dist.irecv, peer, rank + 1))
        for r in (dist.batch_isend_irecv(ops) if ops else []):
            r.wait()
        out = torch.empty((band.out_rows, W - K + 1))
        shard.rowband_conv2d_single_p2p(buf, peer, f, band, out, compute_halo=_oracle_compute_halo,
                                        compute=_oracle_compute)
        np.save(os.path.join(tmpdir, f"band{rank}.npy"), out.numpy())
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,K", [(2, 5), (3, 15), (2, 1)])
def test_rowband_p2p_halo_gloo(world, K):
    import oracle

    H, W = 64, 37
    with tempfile.TemporaryDirectory() as tmp:
        mp.spawn(_worker_rowband_p2p, args=(world, _free_port(), H, W, K, tmp), nprocs=world, join=True)
        got = np.concatenate([np.load(os.path.join(tmp, f"band{r}.npy")) for r in range(world)])
    x = synth.fill_np(11, synth.TAG_INPUT, (H, W), "img")
    ref, _, _ = oracle.conv2d_single(x, synth.make_filter(11, K, "rand")[0, 0])
    assert np.array_equal(got, ref)


def _worker_batch(rank, world, port, tmpdir):
    import oracle

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        N, C, H, W, F, K = 5, 3, 12, 14, 4, 3
        n0, n1 = shard.batch_range(N, world, rank)
        x = synth.fill_np(12, synth.TAG_INPUT, (n1 - n0, C, H, W), "sym", start=n0 * C * H * W)
        w = synth.make_filter(12, K, "he", F=F, C=C)
        yb, _, _ = oracle.conv2d_multi(x, w)
        f0, f1 = shard.filter_range(F, world, rank)
        xa = synth.fill_np(12, synth.TAG_INPUT, (N, C, H, W), "sym")
        yf, _, _ = oracle.conv2d_multi(xa, w[f0:f1])
        # gather across ranks (no collective exists on the data path; this is the test's check)
        gb = [None] * world
        gf = [None] * world
        dist.all_gather_object(gb, yb)
        dist.all_gather_object(gf, yf)
        if rank == 0:
            np.save(os.path.join(tmpdir, "batch.npy"), np.concatenate(gb, axis=0))
            np.save(os.path.join(tmpdir, "filt.npy"), np.concatenate(gf, axis=1))
    finally:
        dist.destroy_process_group()


def test_batch_and_filter_shard_gloo():
    import oracle

    with tempfile.TemporaryDirectory() as tmp:
        mp.spawn(_worker_batch, args=(2, _free_port(), tmp), nprocs=2, join=True)
        xa = synth.fill_np(12, synth.TAG_INPUT, (5, 3, 12, 14), "sym")
        ref, _, _ = oracle.conv2d_multi(xa, synth.make_filter(12, 3, "he", F=4, C=3))
        assert np.array_equal(np.load(os.path.join(tmp, "batch.npy")), ref)
        assert np.array_equal(np.load(os.path.join(tmp, "filt.npy")), ref)

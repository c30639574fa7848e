"""Row-band decomposition across PROCESSES on the device (S 8(e), N3): ranks share one GPU, the band
buffers are exchanged as CUDA IPC mappings (shard.ipc_band_buffers -- on a multi-GPU node the same
call maps a neighbour GPU's memory over NVLink), and every rank computes its band in one
conv2d_single_halo launch reading the neighbour's first K-1 rows in place. The concatenated bands
must equal the one-process conv2d_single bit for bit, and every output must pass the oracle.

The exchange-step path (shard.rowband_conv2d_single: interior call while the K-1 halo rows are in
flight, then the tail call) runs here with the CUDA kernels as `compute` and the halo exchanged over
gloo (NCCL refuses two ranks on one GPU; on a multi-GPU node the same function moves the rows with
NCCL P2P over NVLink)."""
import os
import socket
import tempfile

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from tests.gpu_helpers import check_full_single_host

pytestmark = pytest.mark.gpu


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, H, W, K, out_dir):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    torch.cuda.set_device(0)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from gen import synth
        from paper_conf_cluster_luzw20_b200 import shard

        band = shard.row_band(H, W, K, world, rank)
        buf, peer, keep = shard.ipc_band_buffers(band, torch.device("cuda", 0))
        buf.copy_(synth.fill_torch(synth.BASE_SEED, synth.TAG_INPUT, (band.in_rows, W), "img",
                                   start=band.o0 * W, device="cuda"))
        torch.cuda.synchronize()
        dist.barrier()  # every neighbour's rows are written before anyone reads them in place
        f = torch.from_numpy(synth.make_filter(synth.BASE_SEED, K, "gauss")[0, 0]).cuda()
        out = torch.empty((band.out_rows, W - K + 1), device="cuda")
        shard.rowband_conv2d_single_p2p(buf, peer, f, band, out)
        torch.cuda.synchronize()
        np.save(os.path.join(out_dir, f"band{rank}.npy"), out.cpu().numpy())
        del peer, keep
        dist.barrier()  # the neighbour has finished reading our rows before we free them
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,H,W,K", [(3, 700, 1030, 7), (2, 300, 2048, 15), (2, 120, 517, 3)])
def test_rowband_ipc_halo_in_place(cuda_device, world, H, W, K):
    import paper_conf_cluster_luzw20_b200 as pkg
    from gen import synth

    with tempfile.TemporaryDirectory() as d:
        mp.spawn(_worker, args=(world, _free_port(), H, W, K, d), nprocs=world, join=True)
        got = np.concatenate([np.load(os.path.join(d, f"band{r}.npy")) for r in range(world)])
    x = synth.fill_torch(synth.BASE_SEED, synth.TAG_INPUT, (H, W), "img", device="cuda")
    f = torch.from_numpy(synth.make_filter(synth.BASE_SEED, K, "gauss")[0, 0]).cuda()
    ref = pkg.conv2d_single(x, f).cpu().numpy()
    assert got.shape == ref.shape
    assert np.array_equal(got, ref)
    check_full_single_host(x.cpu().numpy(), f.cpu().numpy(), got)


def _cuda_compute(x, f, out):
    """shard.rowband_conv2d_single `compute` callback: the CUDA C-ABI call on cuda:0 for host band
    buffers (the gloo transport of this test keeps the band on the host)."""
    import paper_conf_cluster_luzw20_b200 as pkg

    out.copy_(pkg.conv2d_single(x.cuda(), f.cuda()).cpu())


def _worker_exchange(rank, world, port, H, W, K, out_dir):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    torch.cuda.set_device(0)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from gen import synth
        from paper_conf_cluster_luzw20_b200 import shard

        band = shard.row_band(H, W, K, world, rank)
        buf = torch.full((band.buf_rows, W), float("nan"))
        buf[:band.in_rows] = synth.fill_torch(synth.BASE_SEED, synth.TAG_INPUT, (band.in_rows, W), "img",
                                              start=band.o0 * W)
        f = torch.from_numpy(synth.make_filter(synth.BASE_SEED, K, "rand")[0, 0])
        out = torch.empty((band.out_rows, W - K + 1))
        shard.rowband_conv2d_single(buf, f, band, out, compute=_cuda_compute)
        np.save(os.path.join(out_dir, f"band{rank}.npy"), out.numpy())
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,H,W,K", [(3, 700, 1030, 7), (2, 300, 2048, 15), (4, 120, 517, 3),
                                         (2, 64, 300, 1)])
def test_rowband_exchange_cuda_compute_vs_oracle(cuda_device, world, H, W, K):
    """Row bands with the exchange step (interior + tail calls of the CUDA kernels): every output
    against the oracle, and bitwise equal to the one-process call."""
    import paper_conf_cluster_luzw20_b200 as pkg
    from gen import synth

    with tempfile.TemporaryDirectory() as d:
        mp.spawn(_worker_exchange, args=(world, _free_port(), H, W, K, d), nprocs=world, join=True)
        got = np.concatenate([np.load(os.path.join(d, f"band{r}.npy")) for r in range(world)])
    x = synth.fill_torch(synth.BASE_SEED, synth.TAG_INPUT, (H, W), "img", device="cuda")
    f = torch.from_numpy(synth.make_filter(synth.BASE_SEED, K, "rand")[0, 0]).cuda()
    check_full_single_host(x.cpu().numpy(), f.cpu().numpy(), got)
    assert np.array_equal(got, pkg.conv2d_single(x, f).cpu().numpy())

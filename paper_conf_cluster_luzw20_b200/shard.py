"""Multi-GPU partitioning of the hot path.

One process per GPU (torchrun), torch.distributed for the plumbing. The paper is single-GPU; the
partitions below come from BASELINE.json north_star / configs[3..4]:

* batch shard  -- rank p takes images [n0, n1): no collective (outputs are independent).
* filter shard -- rank p takes filters [f0, f1) of every image: no collective.
* row band     -- one image too large for one GPU: rank p owns output rows [o_p, o_{p+1}) and the
                  input rows [o_p, o_{p+1}) (the last rank also the final K-1 rows). The one real
                  exchange step: rank p+1 sends its first K-1 input rows to rank p (NCCL P2P over
                  NVLink, torch.distributed.batch_isend_irecv), received into K-1 spare rows at the
                  end of rank p's band buffer. The interior rows, which need no halo, are computed
                  while the halo is in flight; then a tail call computes the last K-1 output rows
                  from 2(K-1) input rows. Outputs are bitwise equal to a one-GPU run (each output's
                  summation order does not depend on where its rows sit; tests pin this).

Fused halo: with the band buffers in symmetric memory (every rank maps its
neighbours' buffers over NVLink), rank p reads rank p+1's first K-1 rows IN PLACE: one
conv2d_single_halo launch computes the whole band, the halo rows streaming over NVLink inside the
kernel's row fetches -- no exchange step, no tail call (`rowband_conv2d_single_p2p`,
`symmetric_band_buffers`).

`compute` defaults to the CUDA C-ABI call; tests on CPU (gloo) pass the oracle instead -- the
product path itself has no CPU fallback.
"""
from __future__ import annotations

from dataclasses import dataclass

import torch
import torch.distributed as dist


def even_split(n: int, world: int, rank: int) -> tuple[int, int]:
    """[start, end) of rank's share of n items, sizes differing by at most one."""
    base, rem = divmod(n, world)
    start = rank * base + min(rank, rem)
    return start, start + base + (1 if rank < rem else 0)


def batch_range(N: int, world: int, rank: int) -> tuple[int, int]:
    return even_split(N, world, rank)


def filter_range(F: int, world: int, rank: int) -> tuple[int, int]:
    return even_split(F, world, rank)


@dataclass(frozen=True)
class RowBand:
    """Rank p's share of a row-band decomposition of one H x W image with a K x K filter."""
    rank: int
    world: int
    H: int
    W: int
    K: int
    o0: int          # first output row owned
    o1: int          # one past the last output row owned
    in_rows: int     # input rows the rank generates / holds: o1-o0 (+K-1 on the last rank)
    buf_rows: int    # rows of the band buffer: o1-o0+K-1 (spare rows receive the halo)

    @property
    def is_last(self) -> bool:
        return self.rank == self.world - 1

    @property
    def out_rows(self) -> int:
        return self.o1 - self.o0

    @property
    def halo(self) -> int:
        return self.K - 1


def row_band(H: int, W: int, K: int, world: int, rank: int) -> RowBand:
    Ho = H - K + 1
    if Ho < world * max(K - 1, 1):
        raise ValueError(f"row bands need at least K-1 = {K - 1} output rows per rank (Ho={Ho}, world={world})")
    o0, o1 = even_split(Ho, world, rank)
    last = rank == world - 1
    in_rows = (o1 - o0) + (K - 1 if last else 0)
    return RowBand(rank, world, H, W, K, o0, o1, in_rows, (o1 - o0) + K - 1)


def _default_compute(x: torch.Tensor, f: torch.Tensor, out: torch.Tensor) -> None:
    from .api import conv2d_single

    conv2d_single(x, f, out=out)


def halo_exchange_ops(buf: torch.Tensor, band: RowBand, group=None):
    """P2P ops of the one exchange step: send my first K-1 rows to rank-1, receive K-1 rows from
    rank+1 into my spare rows. Returns the list of torch.distributed.P2POp."""
    h = band.halo
    ops = []
    if h == 0:
        return ops
    rows = band.out_rows
    if band.rank > 0:
        ops.append(dist.P2POp(dist.isend, buf[:h], band.rank - 1, group))
    if not band.is_last:
        ops.append(dist.P2POp(dist.irecv, buf[rows:rows + h], band.rank + 1, group))
    return ops


def rowband_conv2d_single(buf: torch.Tensor, f: torch.Tensor, band: RowBand, out: torch.Tensor,
                          group=None, compute=_default_compute) -> torch.Tensor:
    """Row-band convolution of rank `band.rank`'s share.

    buf: (band.buf_rows, W) tensor whose first band.in_rows rows hold this rank's input rows
         (the remaining K-1 rows of a non-last rank are overwritten by the halo).
    out: (band.out_rows, W-K+1) output rows [o0, o1) of the full image.
    """
    K, h, rows = band.K, band.halo, band.out_rows
    assert buf.shape[0] == band.buf_rows and out.shape[0] == rows
    ops = halo_exchange_ops(buf, band, group)
    reqs = dist.batch_isend_irecv(ops) if ops else []
    if band.is_last or h == 0:
        # no halo needed: all rows are local (the last rank owns the final K-1 input rows)
        compute(buf[:rows + h], f, out)
        for r in reqs:
            r.wait()
        return out
    interior = rows - h  # output rows computable from own rows alone: [o0, o1-K+1)
    if interior > 0:
        compute(buf[:rows], f, out[:interior])
    for r in reqs:
        r.wait()
    # tail: output rows [o1-K+1, o1) from input rows [o1-K+1, o1+K-1): K-1 own + K-1 halo rows
    t0 = max(interior, 0)
    compute(buf[t0:rows + h], f, out[t0:])
    return out


def _default_compute_halo(x: torch.Tensor, halo: torch.Tensor, f: torch.Tensor, out: torch.Tensor) -> None:
    from .api import conv2d_single_halo

    conv2d_single_halo(x, halo, f, out=out)


def symmetric_band_buffers(band: RowBand, device, group=None):
    """Allocate this rank's band buffer in symmetric memory and map rank+1's first K-1 rows.

    Returns (buf, peer_halo, handle): buf is (band.in_rows, W) local memory every rank can map;
    peer_halo is a (K-1, W) view of rank+1's buf in this device's address space (None on the last
    rank); handle is the symmetric-memory handle (handle.barrier() orders a neighbour's writes before
    our reads). Needs CUDA peer access between the ranks' GPUs (NVLink / NVSwitch)."""
    import torch.distributed._symmetric_memory as symm_mem

    group = group or dist.group.WORLD
    buf = symm_mem.empty((band.in_rows, band.W), dtype=torch.float32, device=device)
    handle = symm_mem.rendezvous(buf, group.group_name)
    peer = None
    if not band.is_last and band.halo > 0:
        peer = handle.get_buffer(band.rank + 1, (band.halo, band.W), torch.float32)
    return buf, peer, handle


def ipc_band_buffers(band: RowBand, device, group=None):
    """Same contract as symmetric_band_buffers, transported by CUDA IPC: every rank allocates its band
    buffer, the IPC handles are exchanged over the process group (all_gather_object), and rank p
    opens rank p+1's buffer in its own address space (lazy peer access over NVLink when the ranks
    are on different GPUs; a plain IPC mapping when they share one -- which lets one GPU test the
    in-place halo path across processes). Returns (buf, peer_halo, keepalive)."""
    from torch.multiprocessing.reductions import reduce_tensor

    buf = torch.empty((band.in_rows, band.W), dtype=torch.float32, device=device)
    handles = [None] * band.world
    dist.all_gather_object(handles, reduce_tensor(buf), group=group)
    peer = None
    if not band.is_last and band.halo > 0:
        rebuild, args = handles[band.rank + 1]
        peer = rebuild(*args)[:band.halo]
    return buf, peer, handles


def rowband_conv2d_single_p2p(buf: torch.Tensor, peer_halo, f: torch.Tensor, band: RowBand, out: torch.Tensor,
                              compute_halo=_default_compute_halo, compute=_default_compute) -> torch.Tensor:
    """Row-band convolution with the halo read in place from the neighbour (one launch per rank).

    buf: (>= band.in_rows, W) this rank's input rows; peer_halo: the first K-1 input rows of rank+1
    (a peer-memory view from symmetric_band_buffers, or any (K-1, W) tensor holding them); ignored on
    the last rank. The caller orders the neighbour's writes of those rows before this call (e.g.
    handle.barrier()); the rows must stay unchanged until the kernel completes.
    out: (band.out_rows, W-K+1) output rows [o0, o1)."""
    rows, h = band.out_rows, band.halo
    assert out.shape[0] == rows
    if band.is_last or h == 0:
        compute(buf[:rows + h], f, out)
    else:
        compute_halo(buf[:rows], peer_halo, f, out)
    return out

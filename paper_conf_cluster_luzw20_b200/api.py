"""Tensor-level API over the C ABI (PyTorch supplies device memory and streams only).

    out = conv2d_single(x, f)      # x: (H, W) fp32 CUDA, f: (K, K)      -> (H-K+1, W-K+1)
    out = conv2d_multi(x, w)       # x: (N, C, H, W), w: (F, C, K, K)    -> (N, F, H-K+1, W-K+1)

Every step of the computation runs in libconv2d.so's kernels; this module only checks types and
shapes, allocates the output, and passes raw pointers plus the current stream. There is no CPU or
eager-PyTorch fallback: non-CUDA tensors raise.

`conv2d_single_host` / `conv2d_multi_host` are the end-to-end entry points for host-resident data:
pinned host -> HBM copy, the kernel, HBM -> host copy, all on one stream (bench.py's `e2e`).
"""
from __future__ import annotations

import torch

from . import _capi


_raw_stream = torch._C._cuda_getCurrentRawStream  # current stream handle of a device index (no Stream object)


def _stream_handle(stream, device_index: int) -> int:
    if stream is None:
        return _raw_stream(device_index)
    return int(stream.cuda_stream)


class _on_device:
    """`with torch.cuda.device(i)` only when i is not already current (the context manager costs
    several microseconds per call, which is most of a small convolution's host time)."""
    __slots__ = ("idx", "prev")

    def __init__(self, idx: int):
        self.idx = idx
        self.prev = -1

    def __enter__(self):
        cur = torch.cuda.current_device()
        if cur != self.idx:
            self.prev = cur
            torch.cuda.set_device(self.idx)

    def __exit__(self, *exc):
        if self.prev >= 0:
            torch.cuda.set_device(self.prev)


def _check_dev(t: torch.Tensor, name: str):
    if not isinstance(t, torch.Tensor):
        raise TypeError(f"{name} must be a torch.Tensor")
    if not t.is_cuda:
        raise TypeError(f"{name} must be a CUDA tensor (no CPU fallback exists)")
    if t.dtype != torch.float32:
        raise TypeError(f"{name} must be float32, got {t.dtype}")
    if not t.is_contiguous():
        raise ValueError(f"{name} must be contiguous")


def _out_for(out, shape, like: torch.Tensor, name="out") -> torch.Tensor:
    """The caller's `out` checked against the result shape (device, dtype, contiguity, same device as
    the input) -- the C ABI cannot know the size of an output buffer -- or a new tensor."""
    shape = tuple(int(v) for v in shape)
    if out is None:
        return torch.empty(shape, dtype=torch.float32, device=like.device)
    _check_dev(out, name)
    if out.device != like.device:
        raise ValueError(f"{name} must be on {like.device}, got {out.device}")
    if tuple(out.shape) != shape:
        raise ValueError(f"{name} has shape {tuple(out.shape)}, expected {shape}")
    return out


def _check_same_device(*ts):
    d = ts[0].device
    for t in ts[1:]:
        if t.device != d:
            raise ValueError(f"all tensors must be on one device ({d} vs {t.device})")


def conv2d_single(x: torch.Tensor, f: torch.Tensor, out: torch.Tensor | None = None, stream=None,
                  band_h: int = 0) -> torch.Tensor:
    _check_dev(x, "x")
    _check_dev(f, "f")
    if x.dim() != 2 or f.dim() != 2 or f.shape[0] != f.shape[1]:
        raise ValueError("x must be (H, W) and f (K, K)")
    _check_same_device(x, f)
    H, W = x.shape
    K = f.shape[0]
    out = _out_for(out, (max(H - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        rc = _capi.lib().conv2d_single_ex(x.data_ptr(), H, W, f.data_ptr(), K, out.data_ptr(),
                                          _stream_handle(stream, dev), band_h)
    if rc:
        _capi.check(rc)
    return out


def conv2d_single_batch(x: torch.Tensor, f: torch.Tensor, out: torch.Tensor | None = None,
                        stream=None) -> torch.Tensor:
    """A batch of images (N, H, W) filtered with one filter f (K, K) in one launch -> (N, H-K+1, W-K+1);
    bitwise equal to conv2d_single on every image. include/conv2d.h: conv2d_single_batch."""
    _check_dev(x, "x")
    _check_dev(f, "f")
    if x.dim() != 3 or f.dim() != 2 or f.shape[0] != f.shape[1]:
        raise ValueError("x must be (N, H, W) and f (K, K)")
    _check_same_device(x, f)
    N, H, W = x.shape
    K = f.shape[0]
    out = _out_for(out, (N, max(H - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        rc = _capi.lib().conv2d_single_batch(x.data_ptr(), N, H, W, f.data_ptr(), K, out.data_ptr(),
                                             _stream_handle(stream, dev))
    if rc:
        _capi.check(rc)
    return out


def conv2d_single_rect(x: torch.Tensor, f: torch.Tensor, out: torch.Tensor | None = None,
                       stream=None) -> torch.Tensor:
    """Valid cross-correlation with a rectangular filter f (FH, FW) -> (H-FH+1, W-FW+1)
    (include/conv2d.h conv2d_single_rect)."""
    _check_dev(x, "x")
    _check_dev(f, "f")
    if x.dim() != 2 or f.dim() != 2:
        raise ValueError("x must be (H, W) and f (FH, FW)")
    _check_same_device(x, f)
    H, W = x.shape
    FH, FW = f.shape
    out = _out_for(out, (max(H - FH + 1, 0), max(W - FW + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        _capi.check(_capi.conv2d_single_rect(x.data_ptr(), H, W, f.data_ptr(), FH, FW, out.data_ptr(),
                                             _stream_handle(stream, dev)))
    return out


def conv2d_single_halo(x: torch.Tensor, halo: torch.Tensor, f: torch.Tensor, out: torch.Tensor | None = None,
                       stream=None) -> torch.Tensor:
    """conv2d_single of the rows of x followed by the rows of halo (same width), without concatenating
    them: the kernels read the halo rows where they are -- e.g. a peer GPU's band buffer mapped over
    NVLink (symmetric memory) -- so a row band is one launch. Bitwise equal to
    conv2d_single(torch.cat([x, halo])). include/conv2d.h: conv2d_single_halo."""
    _check_dev(x, "x")
    _check_dev(halo, "halo")
    _check_dev(f, "f")
    if x.dim() != 2 or halo.dim() != 2 or halo.shape[1] != x.shape[1] or f.dim() != 2 or f.shape[0] != f.shape[1]:
        raise ValueError("x must be (H, W), halo (Hh, W) and f (K, K)")
    H, W = x.shape
    Hh = halo.shape[0]
    K = f.shape[0]
    _check_same_device(x, f)
    out = _out_for(out, (max(H + Hh - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        _capi.check(_capi.conv2d_single_halo(x.data_ptr(), H, W, halo.data_ptr() if Hh else 0, Hh, f.data_ptr(), K,
                                             out.data_ptr(), _stream_handle(stream, dev)))
    return out


_PAD_MODES = {"valid": 0, "same": _capi.CONV2D_PAD_ZERO, "same_zero": _capi.CONV2D_PAD_ZERO,
              "same_replicate": _capi.CONV2D_PAD_REPLICATE}


def conv2d_single_pad(x: torch.Tensor, f: torch.Tensor, padding: str = "same", flip: bool = False,
                      out: torch.Tensor | None = None, stream=None) -> torch.Tensor:
    """Boundary / semantic variants (include/conv2d.h conv2d_single_pad): padding "valid", "same" (=
    "same_zero") or "same_replicate"; flip=True for true convolution (rotated filter)."""
    _check_dev(x, "x")
    _check_dev(f, "f")
    if x.dim() != 2 or f.dim() != 2 or f.shape[0] != f.shape[1]:
        raise ValueError("x must be (H, W) and f (K, K)")
    if padding not in _PAD_MODES:
        raise ValueError(f"padding must be one of {sorted(_PAD_MODES)}")
    mode = _PAD_MODES[padding] | (_capi.CONV2D_FLIP if flip else 0)
    _check_same_device(x, f)
    H, W = x.shape
    K = f.shape[0]
    out = _out_for(out, (H, W) if mode & 3 else (max(H - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        _capi.check(_capi.conv2d_single_pad(x.data_ptr(), H, W, f.data_ptr(), K, mode, out.data_ptr(),
                                            _stream_handle(stream, dev)))
    return out


def conv2d_single_direct(x: torch.Tensor, f: torch.Tensor, out: torch.Tensor | None = None,
                         stream=None) -> torch.Tensor:
    """PAPER.md Fig. 1a baseline kernel (no column/row reuse); evidence control only."""
    _check_dev(x, "x")
    _check_dev(f, "f")
    if x.dim() != 2 or f.dim() != 2 or f.shape[0] != f.shape[1]:
        raise ValueError("x must be (H, W) and f (K, K)")
    _check_same_device(x, f)
    H, W = x.shape
    K = f.shape[0]
    out = _out_for(out, (max(H - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        _capi.check(_capi.conv2d_single_direct(x.data_ptr(), H, W, f.data_ptr(), K, out.data_ptr(),
                                               _stream_handle(stream, dev)))
    return out


def conv2d_multi(x: torch.Tensor, w: torch.Tensor, out: torch.Tensor | None = None, stream=None,
                 band_h: int = 0) -> torch.Tensor:
    _check_dev(x, "x")
    _check_dev(w, "w")
    if x.dim() != 4 or w.dim() != 4 or w.shape[1] != x.shape[1] or w.shape[2] != w.shape[3]:
        raise ValueError("x must be (N, C, H, W) and w (F, C, K, K)")
    _check_same_device(x, w)
    N, C, H, W = x.shape
    F, _, K, _ = w.shape
    out = _out_for(out, (N, F, max(H - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        rc = _capi.lib().conv2d_multi_ex(x.data_ptr(), N, C, H, W, w.data_ptr(), F, K, out.data_ptr(),
                                         _stream_handle(stream, dev), band_h)
    if rc:
        _capi.check(rc)
    return out


def conv2d_multi_tc(x: torch.Tensor, w: torch.Tensor, out: torch.Tensor | None = None, stream=None) -> torch.Tensor:
    """Tensor-core (tcgen05, 3xTF32) variant of conv2d_multi for the large-C dense contraction."""
    _check_dev(x, "x")
    _check_dev(w, "w")
    if x.dim() != 4 or w.dim() != 4 or w.shape[1] != x.shape[1] or w.shape[2] != w.shape[3]:
        raise ValueError("x must be (N, C, H, W) and w (F, C, K, K)")
    _check_same_device(x, w)
    N, C, H, W = x.shape
    F, _, K, _ = w.shape
    out = _out_for(out, (N, F, max(H - K + 1, 0), max(W - K + 1, 0)), x)
    dev = x.device.index
    with _on_device(dev):
        _capi.check(_capi.conv2d_multi_tc(x.data_ptr(), N, C, H, W, w.data_ptr(), F, K, out.data_ptr(),
                                          _stream_handle(stream, dev)))
    return out


def conv2d_single_host(x_host: torch.Tensor, f_host: torch.Tensor, device="cuda", stream=None,
                       out_host: torch.Tensor | None = None, chunk_rows: int = 0) -> torch.Tensor:
    """End-to-end call on host tensors through the C ABI's pipelined host-buffer entry
    (conv2d_single_host): chunked H2D / kernel / D2H overlap. Pin the tensors for full PCIe speed.
    Returns out_host; the result is ready once `stream` (default: the current stream) is synchronised."""
    if x_host.is_cuda or f_host.is_cuda:
        raise TypeError("conv2d_single_host takes host tensors")
    if x_host.dtype != torch.float32 or f_host.dtype != torch.float32:
        raise TypeError("float32 tensors required")
    if x_host.dim() != 2 or f_host.dim() != 2 or f_host.shape[0] != f_host.shape[1]:
        raise ValueError("x_host must be (H, W) and f_host (K, K)")
    x_host = x_host.contiguous()
    f_host = f_host.contiguous()
    H, W = x_host.shape
    K = f_host.shape[0]
    shape = (max(H - K + 1, 0), max(W - K + 1, 0))
    if out_host is None:
        out_host = torch.empty(shape, dtype=torch.float32, pin_memory=True)
    else:
        if out_host.is_cuda or out_host.dtype != torch.float32 or not out_host.is_contiguous():
            raise TypeError("out_host must be a contiguous float32 host tensor")
        if tuple(out_host.shape) != shape:
            raise ValueError(f"out_host has shape {tuple(out_host.shape)}, expected {shape}")
    dev = torch.device(device)
    s = stream if stream is not None else torch.cuda.current_stream(dev)
    with torch.cuda.device(dev):
        _capi.check(_capi.conv2d_single_host(x_host.data_ptr(), H, W, f_host.data_ptr(), K, out_host.data_ptr(),
                                             int(s.cuda_stream), chunk_rows))
    return out_host


def conv2d_multi_host(x_host: torch.Tensor, w_host: torch.Tensor, device="cuda", stream=None,
                      out_host: torch.Tensor | None = None, impl: str = "cuda") -> torch.Tensor:
    """Host tensors in and out around conv2d_multi (impl="cuda", CUDA cores) or conv2d_multi_tc
    (impl="tc", tensor cores), all on one stream."""
    if impl not in ("cuda", "tc"):
        raise ValueError("impl must be 'cuda' or 'tc'")
    dev = torch.device(device)
    s = stream if stream is not None else torch.cuda.current_stream(dev)
    with torch.cuda.stream(s):
        x = x_host.to(dev, non_blocking=True)
        w = w_host.to(dev, non_blocking=True)
        y = (conv2d_multi_tc if impl == "tc" else conv2d_multi)(x, w, stream=s)
        if out_host is None:
            out_host = torch.empty(y.shape, dtype=torch.float32, pin_memory=True)
        out_host.copy_(y, non_blocking=True)
    return out_host

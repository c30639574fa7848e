"""Shared helpers of the GPU parity tests: seeded inputs on the device, oracle checks of full
outputs and of sampled outputs (the oracle recomputes sampled points one by one from patches
gathered out of the device input)."""
from __future__ import annotations

import numpy as np
import torch

import oracle
from gen import synth

TOL = 1e-5  # BASELINE.json north_star: |gpu - ref| <= 1e-5 * sum|x||w|


def dev_image(shape, dist="img", seed=synth.BASE_SEED, device="cuda"):
    return synth.fill_torch(seed, synth.TAG_INPUT, shape, dist, device=device)


def check_full_single(x: torch.Tensor, f: torch.Tensor, y: torch.Tensor, exact: bool = False):
    check_full_single_host(x.cpu().numpy(), f.cpu().numpy(), y.cpu().numpy(), exact)


def check_full_single_host(xh: np.ndarray, fh: np.ndarray, yh: np.ndarray, exact: bool = False):
    """Every output of yh (host copy of the device result) against the oracle on the same input."""
    ref, bound, _ = oracle.conv2d_single(xh, fh)
    assert yh.shape == ref.shape
    if exact:
        bad = ~((yh == ref) | (np.isnan(yh) & np.isnan(ref)))
    else:
        bad = ~oracle.within_tolerance(yh, ref, bound, TOL)
    if bad.any():
        idx = np.argwhere(bad)[:5]
        raise AssertionError(f"{int(bad.sum())} / {bad.size} outputs off; first {idx.tolist()}: "
                             f"gpu {yh[tuple(idx.T)]} ref {ref[tuple(idx.T)]} bound {bound[tuple(idx.T)]}")


def check_full_multi(x, w, y, exact=False):
    xh, wh, yh = x.cpu().numpy(), w.cpu().numpy(), y.cpu().numpy()
    ref, bound, _ = oracle.conv2d_multi(xh, wh)
    assert yh.shape == ref.shape
    bad = ~((yh == ref)) if exact else ~oracle.within_tolerance(yh, ref, bound, TOL)
    if bad.any():
        idx = np.argwhere(bad)[:5]
        raise AssertionError(f"{int(bad.sum())} / {bad.size} outputs off; first {idx.tolist()}: "
                             f"gpu {yh[tuple(idx.T)]} ref {ref[tuple(idx.T)]}")


def sample_points(Ho, Wo, n, rng, band_h=None):
    """Random points plus every corner / first / last row & column and, if given, the rows on both
    sides of band boundaries."""
    ys = list(rng.integers(0, Ho, n))
    xs = list(rng.integers(0, Wo, n))
    edge_y = [0, 1, Ho - 1, Ho - 2, Ho // 2]
    edge_x = [0, 1, 2, 3, 127, 128, 129, Wo - 1, Wo - 2, Wo - 3, Wo - 4, Wo - 129]
    for yy in edge_y:
        for xx in edge_x:
            if 0 <= yy < Ho and 0 <= xx < Wo:
                ys.append(yy)
                xs.append(xx)
    if band_h:
        for b in range(band_h, Ho, band_h * max(1, (Ho // band_h) // 16)):
            for yy in (b - 1, b):
                ys.append(yy)
                xs.append(int(rng.integers(0, Wo)))
    return np.array(ys, np.int64), np.array(xs, np.int64)


def check_points_single(x: torch.Tensor, f: torch.Tensor, y: torch.Tensor, ys, xs):
    """Oracle at sampled outputs: gather each point's K x K input patch from the device input and let
    the oracle compute the point one by one (as a batch of 1x1 outputs)."""
    K = f.shape[0]
    dev = x.device
    yt = torch.as_tensor(ys, device=dev)
    xt = torch.as_tensor(xs, device=dev)
    ar = torch.arange(K, device=dev)
    rows = (yt[:, None] + ar[None, :])[:, :, None]
    cols = (xt[:, None] + ar[None, :])[:, None, :]
    patches = x[rows, cols].cpu().numpy()  # P x K x K
    ref, bound = oracle.conv2d_single_points(patches.reshape(-1, K), f.cpu().numpy(),
                                             np.arange(len(ys)) * K, np.zeros(len(ys), np.int64))
    got = y[yt, xt].cpu().numpy()
    bad = ~oracle.within_tolerance(got, ref, bound, TOL)
    if bad.any():
        i = np.argwhere(bad)[:5, 0]
        raise AssertionError(f"{int(bad.sum())} sampled outputs off: at {list(zip(ys[i], xs[i]))} "
                             f"gpu {got[i]} ref {ref[i]}")


def check_points_multi(x, w, y, ns, fs, ys, xs):
    N, C, H, W = x.shape
    F, _, K, _ = w.shape
    dev = x.device
    nt, yt, xt = (torch.as_tensor(a, device=dev) for a in (ns, ys, xs))
    ar = torch.arange(K, device=dev)
    rows = (yt[:, None] + ar[None, :])[:, None, :, None]
    cols = (xt[:, None] + ar[None, :])[:, None, None, :]
    ch = torch.arange(C, device=dev)[None, :, None, None]
    patches = x[nt[:, None, None, None], ch, rows, cols].cpu().numpy()  # P x C x K x K
    P = len(ns)
    # oracle on a batch of P "images" of size K x K, with each point's own filter
    wh = w.cpu().numpy()
    ref = np.empty(P, np.float32)
    bound = np.empty(P, np.float64)
    fs = np.asarray(fs)
    for f in np.unique(fs):
        sel = np.nonzero(fs == f)[0]
        r, b = oracle.conv2d_multi_points(patches[sel], wh[f:f + 1], np.arange(len(sel)),
                                          np.zeros(len(sel), np.int64), np.zeros(len(sel), np.int64),
                                          np.zeros(len(sel), np.int64))
        ref[sel] = r
        bound[sel] = b
    got = y[nt, torch.as_tensor(fs, device=dev), yt, xt].cpu().numpy()
    bad = ~oracle.within_tolerance(got, ref, bound, TOL)
    if bad.any():
        i = np.argwhere(bad)[:5, 0]
        raise AssertionError(f"{int(bad.sum())} sampled outputs off: gpu {got[i]} ref {ref[i]}")

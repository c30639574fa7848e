"""Seeded, counter-based synthetic input generator (shared by the oracle side and the CUDA side).

This module holds NONE of the convolution's arithmetic: it only turns (seed, tensor tag, global
element index) into fp32 values. Both the CPU oracle (tests, bench cpu_baseline) and the CUDA path
(tests, bench, smoke) draw their inputs from here, so that the two sides see bit-identical data.

Generator:
    h(seed, tag, idx) = splitmix64(seed ^ (tag * PHI64) ^ idx)          (all arithmetic mod 2**64)
    u                 = (h >> 40) * 2**-24                                 exact fp32 in [0, 1)
Distributions of an image / input tensor:
    "img"  u            pixel-like, all-positive (worst case for the 1e-5*sum|x||w| tolerance)
    "sym"  2u - 1       zero-mean, exact in fp32
    "int"  ((h>>40) mod 17) - 8     integers in [-8, 8]  (every fp32 partial sum is exact)
Filters (small, always generated on the host in float64 then rounded once to fp32):
    "rand" (2u - 1) / K          "int"  ((h>>40) mod 9) - 4 in [-4, 4]
    "gauss" sigma = K/6, normalised to sum 1      "box" all ones     "delta" e_(K//2, K//2)
    "he"   N(0, 2/(C*K*K)) by Box-Muller on two uniforms

Because the index is GLOBAL (flat NCHW / row-major index of the full tensor), any shard (batch slice,
row band) can be generated independently and matches the single-GPU tensor bit for bit.

Two bit-identical implementations: numpy uint64 (host) and torch int64 (any device, used to fill
large images directly in HBM). tests/test_gen.py pins them against each other and against the
published splitmix64 test vector.
"""
from __future__ import annotations

import math

import numpy as np

PHI64 = 0x9E3779B97F4A7C15
_M1 = 0xBF58476D1CE4E5B9
_M2 = 0x94D049BB133111EB
_MASK64 = (1 << 64) - 1

BASE_SEED = 20200914  # Cluster 2020 opening day; config index is added per config

TAG_INPUT = 1
TAG_FILTER = 2

IMAGE_DISTS = ("img", "sym", "int")
FILTER_DISTS = ("rand", "int", "gauss", "box", "delta", "he")


# ----------------------------------------------------------------------------------------------
# numpy (host) implementation
# ----------------------------------------------------------------------------------------------
def splitmix64_np(x: np.ndarray) -> np.ndarray:
    """splitmix64 finaliser of (x + PHI64); x is uint64. Wraps mod 2**64."""
    with np.errstate(over="ignore"):
        z = x.astype(np.uint64) + np.uint64(PHI64)
        z = (z ^ (z >> np.uint64(30))) * np.uint64(_M1)
        z = (z ^ (z >> np.uint64(27))) * np.uint64(_M2)
        return z ^ (z >> np.uint64(31))


def _key(seed: int, tag: int) -> int:
    return (int(seed) ^ ((int(tag) * PHI64) & _MASK64)) & _MASK64


def hash_np(seed: int, tag: int, start: int, n: int) -> np.ndarray:
    idx = np.arange(start, start + n, dtype=np.uint64)
    return splitmix64_np(idx ^ np.uint64(_key(seed, tag)))


def _from_hash_np(h: np.ndarray, dist: str) -> np.ndarray:
    top = (h >> np.uint64(40)).astype(np.int64)  # 24 random bits
    if dist == "img":
        return (top.astype(np.float32) * np.float32(2.0 ** -24)).astype(np.float32)
    if dist == "sym":
        return ((top - (1 << 23)).astype(np.float32) * np.float32(2.0 ** -23)).astype(np.float32)
    if dist == "int":
        return ((top % 17) - 8).astype(np.float32)
    raise ValueError(f"unknown image distribution {dist!r}")


def fill_np(seed: int, tag: int, shape, dist: str = "img", start: int = 0,
            chunk: int = 1 << 24) -> np.ndarray:
    """fp32 tensor of `shape` whose flat element e carries global index start+e."""
    n = int(np.prod(shape)) if len(shape) else 1
    out = np.empty(n, dtype=np.float32)
    for s in range(0, n, chunk):
        m = min(chunk, n - s)
        out[s:s + m] = _from_hash_np(hash_np(seed, tag, start + s, m), dist)
    return out.reshape(shape)


# ----------------------------------------------------------------------------------------------
# torch implementation (int64 two's-complement emulation of the same uint64 arithmetic)
# ----------------------------------------------------------------------------------------------
def _s64(v: int) -> int:
    v &= _MASK64
    return v - (1 << 64) if v >= (1 << 63) else v


def _lsr(z, s: int):
    """logical right shift of an int64 tensor holding uint64 bits"""
    return (z >> s) & ((1 << (64 - s)) - 1)


def fill_torch(seed: int, tag: int, shape, dist: str = "img", start: int = 0, device="cpu",
               chunk: int = 1 << 26):
    """Same values as fill_np, produced on `device` (e.g. straight into HBM)."""
    import torch

    n = 1
    for d in shape:
        n *= int(d)
    out = torch.empty(n, dtype=torch.float32, device=device)
    key = _s64(_key(seed, tag))
    for s in range(0, n, chunk):
        m = min(chunk, n - s)
        z = torch.arange(start + s, start + s + m, dtype=torch.int64, device=device)
        z ^= key
        z += _s64(PHI64)
        z = (z ^ _lsr(z, 30)) * _s64(_M1)
        z = (z ^ _lsr(z, 27)) * _s64(_M2)
        z = z ^ _lsr(z, 31)
        top = _lsr(z, 40)
        if dist == "img":
            out[s:s + m] = top.to(torch.float32) * (2.0 ** -24)
        elif dist == "sym":
            out[s:s + m] = (top - (1 << 23)).to(torch.float32) * (2.0 ** -23)
        elif dist == "int":
            out[s:s + m] = ((top % 17) - 8).to(torch.float32)
        else:
            raise ValueError(f"unknown image distribution {dist!r}")
        del z, top
    return out.reshape(tuple(int(d) for d in shape))


# ----------------------------------------------------------------------------------------------
# filters (host, float64 then one rounding to fp32)
# ----------------------------------------------------------------------------------------------
def _uniform01_f64(seed: int, tag: int, n: int, start: int = 0) -> np.ndarray:
    top = (hash_np(seed, tag, start, n) >> np.uint64(11)).astype(np.float64)  # 53 bits
    return top * 2.0 ** -53


def make_filter(seed: int, K: int, dist: str = "rand", F: int = 1, C: int = 1,
                tag: int = TAG_FILTER) -> np.ndarray:
    """Filter bank of shape (F, C, K, K) (FCKK == torch OIHW) as fp32."""
    n = F * C * K * K
    if dist == "rand":
        h = hash_np(seed, tag, 0, n)
        u = (h >> np.uint64(40)).astype(np.float64) * 2.0 ** -24
        w = (2.0 * u - 1.0) / K
    elif dist == "int":
        h = hash_np(seed, tag, 0, n)
        w = ((h >> np.uint64(40)).astype(np.int64) % 9 - 4).astype(np.float64)
    elif dist == "gauss":
        sig = K / 6.0
        c = (K - 1) / 2.0
        ii, jj = np.meshgrid(np.arange(K), np.arange(K), indexing="ij")
        g = np.exp(-((ii - c) ** 2 + (jj - c) ** 2) / (2.0 * sig * sig))
        g = g / g.sum()
        w = np.broadcast_to(g, (F, C, K, K)).copy()
    elif dist == "box":
        w = np.ones(n, dtype=np.float64)
    elif dist == "delta":
        w = np.zeros((F, C, K, K), dtype=np.float64)
        w[:, :, K // 2, K // 2] = 1.0
    elif dist == "he":
        u1 = _uniform01_f64(seed, tag, n, 0)
        u2 = _uniform01_f64(seed, tag, n, n)
        z = np.sqrt(-2.0 * np.log1p(-u1)) * np.cos(2.0 * math.pi * u2)
        w = z * math.sqrt(2.0 / (C * K * K))
    else:
        raise ValueError(f"unknown filter distribution {dist!r}")
    return np.asarray(w, dtype=np.float64).reshape(F, C, K, K).astype(np.float32)

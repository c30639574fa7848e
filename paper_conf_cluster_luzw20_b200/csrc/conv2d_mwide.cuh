// conv2d_mwide.cuh -- multi-channel kernel with wide lanes (8 contiguous output columns per lane).
//
// The wide single-channel design (conv2d_wide.cuh) extended along the multi-channel axes of PAPER.md's
// multi-channel experiment (Table I), replacing k_conv2d_multi2's 4-column lanes:
//   * a5 channel reduction: for every input row r the C channel rows stream through the same K-slot
//     accumulator ring (the first channel also shifts the ring): each output sums its C*K*K terms in
//     (filter row, channel, filter column) order -- the order of k_conv2d_multi2 (same bits);
//   * FB filters per warp, filters of the CTA's F-block staged in shared memory and read with
//     broadcast LDS.128. A broadcast LDS.128 moves 512 B through the shared-memory crossbar (4 cycles
//     of its 128 B/clk): with 4-column lanes one filter value feeds 4 FMAs per lane and the SM's FMA
//     pipes (4 warp-FFMA/clk) outrun the filter supply (1 value/clk) -- k_conv2d_multi2 is bound there
//     (configs[2] 25%, configs[3] 51% of fp32 peak). With 8 columns per lane a value feeds 8 FMAs:
//     the crossbar runs at ~50% and the FMA pipe can lead;
//   * SEG-lane segments (SEG in {4, 8, 16, 32}): a segment of SEG lanes covers 8*SEG columns of one
//     image, a warp 32/SEG images, so narrow layers keep their lanes busy (Table I: 8-222 columns);
//     the column-reuse shuffles stay inside the segment;
//   * row fetch: each (row, channel) entry's own 8 columns + the halo quads of segment lanes 0/1,
//     one or two entries in flight in registers;
//   * output: SEG = 32 (one image per warp): each lane's 8 outputs realigned to 16-byte quads with
//     shfl.down (the row shift is warp-uniform); SEG < 32: masked scalar stores.
#pragma once

#include <type_traits>

#include "conv2d_multi.cuh"
#include "conv2d_wide.cuh"

namespace c2d {

// a3 + a5: one (row, channel) entry into the ring of FB filters x 8 columns
template <int K, int FB, bool SHIFT, bool GUARD>
__device__ __forceinline__ void mwide_step(float (&acc)[K][FB][kWideV], const float (&w)[WideCfg<K>::WN],
                                           const MultiFilter<K, FB> &mf, int c, int qmin, int qmax) {
#pragma unroll
  for (int q = 0; q < K; ++q) {
    if (!GUARD || (q >= qmin && q < qmax)) {
#pragma unroll
      for (int fb = 0; fb < FB; ++fb) {
        float fr[KCfg<K>::KP];
        mf.row(fr, fb, c, K - 1 - q);
#pragma unroll
        for (int v = 0; v < kWideV; ++v) {
          float s;
          if (SHIFT)
            s = (q + 1 < K) ? acc[(q + 1 < K) ? q + 1 : 0][fb][v] : 0.f;
          else
            s = acc[q][fb][v];
#pragma unroll
          for (int j = 0; j < K; ++j) s = fmaf(w[v + j], fr[j], s);
          acc[q][fb][v] = s;
        }
      }
    }
  }
}

// EDGE 0: interior tile (vector loads; SEG = 32: realigned vector stores); 1: aligned rows, ragged right
// edge (clamped vector loads, masked scalar stores); 2: misaligned rows (guarded scalar loads, masked
// stores). PF: 1 or 2 (row, channel) entries in flight in registers.
template <int K, int FB, int SEG, int GUARDS, int PF, int EDGE>
__device__ __forceinline__ void mwide_tile(const Multi2Args &a, const MultiFilter<K, FB> &mf, int n, bool seg_active,
                                           int f0, int x0, int ob, int oe, int lane) {
  constexpr bool SAFE = (EDGE != 0);
  const int sl = lane & (SEG - 1);
  const int C = a.C;
  const int rend = oe + K - 1;
  const int rlast = rend - 1;
  const size_t plane = static_cast<size_t>(a.H) * a.W;
  const float *__restrict__ img = a.in + static_cast<size_t>(n) * C * plane;
  float acc[K][FB][kWideV];
#pragma unroll
  for (int q = 0; q < K; ++q)
#pragma unroll
    for (int fb = 0; fb < FB; ++fb)
#pragma unroll
      for (int v = 0; v < kWideV; ++v) acc[q][fb][v] = 0.f;

  // the (row, channel) stream: (r, c) -> (r, c+1) -> ... -> (r+1, 0)
  const float *__restrict__ fetch_row0 = img + static_cast<size_t>(ob) * a.W;  // channel 0 of row pr
  const float *__restrict__ fetch = fetch_row0;
  int pr = ob, pc = 0;
  auto advance = [&]() {
    if (++pc == C) {
      pc = 0;
      if (pr < rlast) {
        ++pr;
        fetch_row0 += a.W;
      }
      fetch = fetch_row0;
    } else {
      fetch += plane;
    }
  };
  WideRow n1, n2;
  wide_load<K, EDGE, SEG>(n1, fetch, x0, a.W, sl);
  advance();
  if constexpr (PF == 2) {
    wide_load<K, EDGE, SEG>(n2, fetch, x0, a.W, sl);
    advance();
  }
  auto stream_row = [&](int qmin, int qmax, auto guard_tag) {
    constexpr bool G = decltype(guard_tag)::value;
    for (int c = 0; c < C; ++c) {
      WideRow cur = n1;
      if constexpr (PF == 2) {
        n1 = n2;
        wide_load<K, EDGE, SEG>(n2, fetch, x0, a.W, sl);
      } else {
        wide_load<K, EDGE, SEG>(n1, fetch, x0, a.W, sl);
      }
      advance();
      float w[WideCfg<K>::WN];
      wide_window<K, SEG>(cur, w, lane);
      if (c == 0)
        mwide_step<K, FB, true, G>(acc, w, mf, c, qmin, qmax);
      else
        mwide_step<K, FB, false, G>(acc, w, mf, c, qmin, qmax);
    }
  };
  auto store_slot0 = [&](int o) {
#pragma unroll
    for (int fb = 0; fb < FB; ++fb) {
      const int f = f0 + fb;
      if (f < a.F) {
        float *orow = a.out + ((static_cast<size_t>(n) * a.F + f) * a.Ho + o) * a.Wo;
        if constexpr (SEG == kWarp && !SAFE) {
          wide_store<false>(orow, x0, a.Wo, acc[0][fb], lane);
        } else if (seg_active) {
#pragma unroll
          for (int t = 0; t < kWideV; ++t) {
            const int x = x0 + kWideV * sl + t;
            if (x < a.Wo) __stcs(orow + x, acc[0][fb][t]);
          }
        }
      }
    }
  };
  int r = ob;
  if constexpr (GUARDS == 0) {
    for (; r < rend; ++r) {
      stream_row(0, K, std::false_type{});
      if (r >= ob + K - 1) store_slot0(r - K + 1);
    }
  } else {
    for (; r < min(ob + K - 1, oe); ++r) stream_row(K - 1 - (r - ob), K, std::true_type{});
    for (; r < oe; ++r) {
      stream_row(0, K, std::false_type{});
      store_slot0(r - K + 1);
    }
    for (; r < rend; ++r) {
      stream_row(max(0, K - 1 - (r - ob)), oe + K - 1 - r, std::true_type{});
      if (r >= ob + K - 1) store_slot0(r - K + 1);
    }
  }
}

// Tiles are ordered ((group * n_fb + fblk) * n_bands + band) * n_cb + cb as k_conv2d_multi2 (the host
// pads n_bands so that the CTA's 4 warps share (group, fblk)); the CTA stages that F-block's filters.
template <int K, int FB, int SEG, int GUARDS, int PF, int MINB>
__global__ void __launch_bounds__(kCtaWarps *kWarp, MINB) k_conv2d_mwide(const Multi2Args a) {
  constexpr int KP = KCfg<K>::KP;
  extern __shared__ __align__(16) float smem[];
  const long long tile0 = static_cast<long long>(blockIdx.x) * kCtaWarps;
  const long long per_fb = static_cast<long long>(a.n_cb) * a.n_bands;
  const int fblk = static_cast<int>((tile0 / per_fb) % a.n_fb);
  const int f0 = fblk * FB;
  const int total = a.C * K * FB * KP;
  for (int t = threadIdx.x; t < total; t += blockDim.x) {
    const int j = t % KP;
    const int fb = (t / KP) % FB;
    const int i = (t / (KP * FB)) % K;
    const int c = t / (KP * FB * K);
    const int f = f0 + fb;
    smem[t] = (j < K && f < a.F) ? a.filt[((static_cast<size_t>(f) * a.C + c) * K + i) * K + j] : 0.f;
  }
  __syncthreads();
  MultiFilter<K, FB> mf;
  mf.sbase = static_cast<unsigned>(__cvta_generic_to_shared(smem));
  const int lane = threadIdx.x & (kWarp - 1);
  const long long tile = tile0 + (threadIdx.x >> 5);
  if (tile >= a.n_tiles) return;
  const int cb = static_cast<int>(tile % a.n_cb);
  const int band = static_cast<int>((tile / a.n_cb) % a.n_bands);
  const int group = static_cast<int>(tile / (per_fb * a.n_fb));
  const int ob = band * a.band_h;
  if (ob >= a.Ho) return;
  const int oe = min(ob + a.band_h, a.Ho);
  const int x0 = cb * kWideV * SEG;
  constexpr int SEGS = kWarp / SEG;
  const int n_raw = group * SEGS + lane / SEG;
  const bool seg_active = n_raw < a.N;
  const int n = seg_active ? n_raw : a.N - 1;  // idle segments recompute the last image, never store
  const bool inside = x0 + kWideV * SEG + 16 <= a.W;  // span + both halo quads (uniform per warp)
  if (a.aligned && inside)
    mwide_tile<K, FB, SEG, GUARDS, PF, 0>(a, mf, n, seg_active, f0, x0, ob, oe, lane);
  else if (a.aligned)
    mwide_tile<K, FB, SEG, GUARDS, PF, 1>(a, mf, n, seg_active, f0, x0, ob, oe, lane);
  else
    mwide_tile<K, FB, SEG, GUARDS, PF, 2>(a, mf, n, seg_active, f0, x0, ob, oe, lane);
}

}  // namespace c2d

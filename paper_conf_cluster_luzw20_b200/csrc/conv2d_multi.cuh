// conv2d_multi.cuh -- multi-channel kernel (N images x C channels x F filters of K x K), sm_100a.
//
// The single-channel design (conv2d_kernels.cuh) extended along the two new axes of PAPER.md's
// multi-channel experiment (Table I):
//   * a5 channel reduction: for every input row r the C channel rows stream through the same K-slot
//     accumulator ring (the first channel also shifts the ring), so each output sums its C*K*K terms
//     in (filter row, channel, filter column) order, band-independent;
//   * FB filters per warp: one assembled window (column reuse) feeds K slots x FB filters x 4 x K FMAs;
//   * SEG-lane segments: a warp is split into 32/SEG segments of SEG lanes (4*SEG columns each) that
//     work on different images n with identical control flow, so narrow images (e.g. the 54-column
//     outputs of 56x56 layers) do not leave most lanes idle. The column-reuse shuffles wrap inside a
//     segment (shfl.idx with a segment-local source lane);
//   * U chunks of 4*SEG columns per segment share every filter-row fetch (more FMAs per LDS);
//   * filters: the CTA's F-block staged in shared memory (4 warps per CTA share it), broadcast LDS.128.
//     (A __constant__ filter bank read through uniform registers -- the single-channel choice -- does
//     not work here: warps on one SM use different F-blocks, the working set overflows the constant
//     cache and LDCU latency serialises the warp; measured 3 vs 24 TFLOP/s on configs[3].)
// Alg. 2's first/last K-1 rows of a band (cases 1 and 3) are guarded per slot (GUARDS=2) when bands
// are short, or run the full body (GUARDS=0) when bands are tall.
#pragma once

#include <type_traits>

#include "conv2d_kernels.cuh"

namespace c2d {

struct Multi2Args {
  const float *in;
  const float *filt;  // F x C x K x K in global memory
  float *out;
  int N, C, H, W, F, Ho, Wo;
  int band_h, n_cb, n_bands, n_fb, n_groups;
  long long n_tiles;
  int aligned;
};

// filter row (fb, c, i) of the CTA's F-block, staged in shared memory as [c][i][fb][KP]
template <int K, int FB>
struct MultiFilter {
  unsigned sbase;

  __device__ __forceinline__ void row(float (&fr)[KCfg<K>::KP], int fb, int c, int i) const {
    constexpr int KP = KCfg<K>::KP;
#pragma unroll
    for (int c4 = 0; c4 < KP / 4; ++c4)
      lds4_at(sbase + static_cast<unsigned>((((c * K + i) * FB + fb) * KP + 4 * c4) * 4), fr[4 * c4],
              fr[4 * c4 + 1], fr[4 * c4 + 2], fr[4 * c4 + 3]);
  }
};

// The F-block staged as [c][i][j][fb] (filters fastest) for the paired-FMA step: one LDS.128 at (c, i, j)
// returns the filter values of four consecutive filters, i.e. two aligned (fb, fb+1) register pairs.
template <int K, int FB>
struct MultiFilterP2 {
  static_assert(FB % 2 == 0, "filter pairs");
  unsigned sbase;
  // fr2[p][j] = (w[f0+2p][c][i][j], w[f0+2p+1][c][i][j])
  __device__ __forceinline__ void row2(float2 (&fr2)[FB / 2][K], int c, int i) const {
#pragma unroll
    for (int j = 0; j < K; ++j) {
      const unsigned base = sbase + static_cast<unsigned>((((c * K + i) * K + j) * FB) * 4);
      if constexpr (FB == 2) {
        float x, y;
        asm volatile("ld.shared.v2.f32 {%0, %1}, [%2];" : "=f"(x), "=f"(y) : "r"(base));
        fr2[0][j] = make_float2(x, y);
      } else {
#pragma unroll
        for (int p = 0; p < FB / 2; p += 2) {
          float a0, a1, a2, a3;
          lds4_at(base + p * 8, a0, a1, a2, a3);
          fr2[p][j] = make_float2(a0, a1);
          fr2[p + 1][j] = make_float2(a2, a3);
        }
      }
    }
  }
};

// a3 + a5 with paired FMA (sm_100 FFMA2): one instruction runs the chains of filters fb and fb+1 at the
// same column -- the window value broadcast (FFMA2's scalar register operand), the filter pair from one
// register pair, the accumulator pair. Same fmaf steps per output as row_step_multi: the same bits.
template <int K, int FB, int U, bool SHIFT, bool GUARD>
__device__ __forceinline__ void row_step_multi_p2(float (&acc)[K][FB][U][4], const float (&w)[U][KCfg<K>::WN],
                                                  const MultiFilterP2<K, FB> &mf, int c, int qmin, int qmax) {
#pragma unroll
  for (int q = 0; q < K; ++q) {
    if (!GUARD || (q >= qmin && q < qmax)) {
      float2 fr2[FB / 2][K];
      mf.row2(fr2, c, K - 1 - q);
#pragma unroll
      for (int p = 0; p < FB / 2; ++p) {
#pragma unroll
        for (int u = 0; u < U; ++u) {
#pragma unroll
          for (int v = 0; v < 4; ++v) {
            const int qs = SHIFT ? ((q + 1 < K) ? q + 1 : 0) : q;
            float2 s = (SHIFT && q + 1 >= K) ? make_float2(0.f, 0.f)
                                              : make_float2(acc[qs][2 * p][u][v], acc[qs][2 * p + 1][u][v]);
#pragma unroll
            for (int j = 0; j < K; ++j) s = __ffma2_rn(make_float2(w[u][v + j], w[u][v + j]), fr2[p][j], s);
            acc[q][2 * p][u][v] = s.x;
            acc[q][2 * p + 1][u][v] = s.y;
          }
        }
      }
    }
  }
}

// a3 + a5: one (row, channel) into the ring of FB filters x U chunks
template <int K, int FB, int U, bool SHIFT, bool GUARD, typename MF>
__device__ __forceinline__ void row_step_multi(float (&acc)[K][FB][U][4], const float (&w)[U][KCfg<K>::WN],
                                               const MF &mf, int c, int qmin, int qmax) {
#pragma unroll
  for (int q = 0; q < K; ++q) {
    if (!GUARD || (q >= qmin && q < qmax)) {
#pragma unroll
      for (int fb = 0; fb < FB; ++fb) {
        float fr[KCfg<K>::KP];
        mf.row(fr, fb, c, K - 1 - q);
#pragma unroll
        for (int u = 0; u < U; ++u) {
#pragma unroll
          for (int v = 0; v < 4; ++v) {
            float s;
            if (SHIFT)
              s = (q + 1 < K) ? acc[(q + 1 < K) ? q + 1 : 0][fb][u][v] : 0.f;
            else
              s = acc[q][fb][u][v];
#pragma unroll
            for (int j = 0; j < K; ++j) s = fmaf(w[u][v + j], fr[j], s);
            acc[q][fb][u][v] = s;
          }
        }
      }
    }
  }
}

// EDGE 0: interior tile (ring, vector stores); 1: aligned rows, ragged right edge (ring with clamped
// addresses, masked scalar stores); 2: misaligned rows (guarded scalar loads in registers, masked stores)
template <int K, int FB, int U, int SEG, int GUARDS, int PF, int EDGE, typename MF>
__device__ __forceinline__ void multi_tile2(const Multi2Args &a, const MF &mf, int n,
                                            bool seg_active, int f0, int x0, int ob, int oe, int lane,
                                            unsigned ring_base) {
  const int sl = lane & (SEG - 1);
  const int C = a.C;
  const int rend = oe + K - 1;
  const int rlast = rend - 1;
  const size_t plane = static_cast<size_t>(a.H) * a.W;
  const float *__restrict__ img = a.in + static_cast<size_t>(n) * C * plane;
  float acc[K][FB][U][4];
#pragma unroll
  for (int q = 0; q < K; ++q)
#pragma unroll
    for (int fb = 0; fb < FB; ++fb)
#pragma unroll
      for (int u = 0; u < U; ++u)
#pragma unroll
        for (int v = 0; v < 4; ++v) acc[q][fb][u][v] = 0.f;

  // the (row, channel) stream: (r, c) -> (r, c+1) -> ... -> (r+1, 0). PF >= 3 and aligned rows: a
  // PF-stage cp.async ring in shared memory (PF-1 entries in flight); otherwise PF (1 or 2) entries
  // in registers (misaligned rows: one).
  constexpr bool SAFE = (EDGE != 0);
  constexpr int NST = (PF >= 3 && EDGE != 2) ? PF : 1;
  constexpr int RPF = (NST == 1 && PF == 2 && EDGE != 2) ? 2 : 1;  // register prefetch depth
  static_assert(NST == 1 || (NST & (NST - 1)) == 0, "ring depth must be a power of two");
  RowRing<K, U, SEG, (NST > 1 ? NST : 2)> ring;
  ring.base = ring_base;
  ring.lane = lane;
  ring.sl = sl;
  RowBuf<K, U> n1, n2;  // register path: PF (1 or 2) entries in flight
  // next entry to fetch: pointer advanced by one channel plane per entry, by one row after C entries
  const float *__restrict__ fetch_row0 = img + static_cast<size_t>(ob) * a.W;  // channel 0 of row pr
  const float *__restrict__ fetch = fetch_row0;
  int pr = ob, pc = 0;
  int t = 0;  // entries consumed
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
  constexpr bool clamp = (EDGE == 1);
  if constexpr (NST > 1) {
#pragma unroll
    for (int st = 0; st < NST - 1; ++st) {
      ring.issue(st, fetch, x0, a.W, clamp);
      advance();
    }
  } else {
    load_row_g<K, U, SEG, SAFE>(n1, fetch, x0, a.W, sl, a.aligned);
    advance();
    if constexpr (RPF == 2) {
      load_row_g<K, U, SEG, SAFE>(n2, fetch, x0, a.W, sl, a.aligned);
      advance();
    }
  }
  auto stream_row = [&](int r, int qmin, int qmax, auto guard_tag) {
    constexpr bool G = decltype(guard_tag)::value;
    for (int c = 0; c < C; ++c) {
      RowBuf<K, U> cur;
      if constexpr (NST > 1) {
        cp_async_wait<NST - 2>();
        ring.read(t & (NST - 1), cur);
        ring.issue((t + NST - 1) & (NST - 1), fetch, x0, a.W, clamp);  // the stage read at t-1
        ++t;
      } else if constexpr (RPF == 2) {
        cur = n1;
        n1 = n2;
        load_row_g<K, U, SEG, SAFE>(n2, fetch, x0, a.W, sl, a.aligned);
      } else {
        cur = n1;
        load_row_g<K, U, SEG, SAFE>(n1, fetch, x0, a.W, sl, a.aligned);
      }
      advance();
      float w[U][KCfg<K>::WN];
      build_windows_g<K, U, SEG>(cur, w, lane);
      if constexpr (std::is_same<MF, MultiFilterP2<K, FB>>::value) {
        if (c == 0)
          row_step_multi_p2<K, FB, U, true, G>(acc, w, mf, c, qmin, qmax);
        else
          row_step_multi_p2<K, FB, U, false, G>(acc, w, mf, c, qmin, qmax);
      } else {
        if (c == 0)
          row_step_multi<K, FB, U, true, G>(acc, w, mf, c, qmin, qmax);
        else
          row_step_multi<K, FB, U, false, G>(acc, w, mf, c, qmin, qmax);
      }
    }
  };
  auto store_slot0 = [&](int o) {
#pragma unroll
    for (int fb = 0; fb < FB; ++fb) {
      const int f = f0 + fb;
      if (f < a.F) {
        float *orow = a.out + ((static_cast<size_t>(n) * a.F + f) * a.Ho + o) * a.Wo;
#pragma unroll
        for (int u = 0; u < U; ++u) {
          const int xb = x0 + 4 * SEG * u;
          if constexpr (SEG == kWarp && !SAFE) {
            store_chunk(orow + xb, acc[0][fb][u], lane);
          } else if (seg_active) {
#pragma unroll
            for (int t = 0; t < 4; ++t) {
              const int x = xb + 4 * sl + t;
              if (x < a.Wo) __stcs(orow + x, acc[0][fb][u][t]);
            }
          }
        }
      }
    }
  };
  int r = ob;
  if constexpr (GUARDS == 0) {
    for (; r < rend; ++r) {
      stream_row(r, 0, K, std::false_type{});
      if (r >= ob + K - 1) store_slot0(r - K + 1);
    }
  } else {
    for (; r < min(ob + K - 1, oe); ++r) stream_row(r, K - 1 - (r - ob), K, std::true_type{});
    for (; r < oe; ++r) {
      stream_row(r, 0, K, std::false_type{});
      store_slot0(r - K + 1);
    }
    for (; r < rend; ++r) {
      stream_row(r, max(0, K - 1 - (r - ob)), oe + K - 1 - r, std::true_type{});
      if (r >= ob + K - 1) store_slot0(r - K + 1);
    }
  }
}

// Tiles are ordered ((group * n_fb + fblk) * n_bands + band) * n_cb + cb; the host pads n_bands so that
// the CTA's warps share (group, fblk): the CTA stages that F-block's C*K*FB*KP floats once.
// MINB: resident CTAs per SM the register allocation is capped for (3: <= 168 registers; whole-warp
// rows with FB = 8 at K <= 3 need more: MINB = 2 there). ALIGNED: the launch's input is 16-byte aligned
// with W % 4 == 0 (interior + ragged-edge tiles); the misaligned case (guarded scalar loads) is its own
// instantiation, so its register demand never caps -- or spills in -- the hot kernel (0 LDL/STL,
// tests/test_sass.py).
// P2: paired FMA across filter pairs (row_step_multi_p2), F-block staged [c][i][j][fb].
template <int K, int FB, int U, int SEG, int GUARDS, int PF, int MINB = 3, bool ALIGNED = true, bool P2 = false>
__global__ void __launch_bounds__(kCtaWarps *kWarp, MINB) k_conv2d_multi2(const Multi2Args a) {
  constexpr int KP = KCfg<K>::KP;
  extern __shared__ __align__(16) float smem[];
  const long long tile0 = static_cast<long long>(blockIdx.x) * kCtaWarps;
  const long long per_fb = static_cast<long long>(a.n_cb) * a.n_bands;
  const int fblk = static_cast<int>((tile0 / per_fb) % a.n_fb);
  const int f0 = fblk * FB;
  const int total = P2 ? a.C * K * K * FB : a.C * K * FB * KP;
  for (int t = threadIdx.x; t < total; t += blockDim.x) {
    int c, i, j, fb;
    if constexpr (P2) {  // [c][i][j][fb]
      fb = t % FB;
      j = (t / FB) % K;
      i = (t / (FB * K)) % K;
      c = t / (FB * K * K);
    } else {  // [c][i][fb][KP]
      j = t % KP;
      fb = (t / KP) % FB;
      i = (t / (KP * FB)) % K;
      c = t / (KP * FB * K);
    }
    const int f = f0 + fb;
    smem[t] = (j < K && f < a.F) ? a.filt[((static_cast<size_t>(f) * a.C + c) * K + i) * K + j] : 0.f;
  }
  __syncthreads();
  using MF = typename std::conditional<P2, MultiFilterP2<K, FB>, MultiFilter<K, FB>>::type;
  MF mf;
  mf.sbase = static_cast<unsigned>(__cvta_generic_to_shared(smem));
  const int lane = threadIdx.x & (kWarp - 1);
  // this warp's cp.async row ring, after the F-block, 16-byte aligned (the P2 layout C*K*K*FB may not be a
  // multiple of 4 floats)
  const unsigned ring_base = mf.sbase + static_cast<unsigned>((total + 3) / 4 * 4) * 4u +
                             (threadIdx.x >> 5) * RowRing<K, U, SEG, (PF >= 3 ? PF : 2)>::kBytes;
  const long long tile = tile0 + (threadIdx.x >> 5);
  if (tile >= a.n_tiles) return;
  const int cb = static_cast<int>(tile % a.n_cb);
  const int band = static_cast<int>((tile / a.n_cb) % a.n_bands);
  const int group = static_cast<int>(tile / (per_fb * a.n_fb));
  const int ob = band * a.band_h;
  if (ob >= a.Ho) return;
  const int oe = min(ob + a.band_h, a.Ho);
  const int x0 = cb * 4 * SEG * U;
  constexpr int SEGS = kWarp / SEG;
  const int n_raw = group * SEGS + lane / SEG;
  const bool seg_active = n_raw < a.N;
  const int n = seg_active ? n_raw : a.N - 1;  // idle segments recompute the last image, never store
  const bool inside = x0 + 4 * SEG * U + 4 * KCfg<K>::NE <= a.W;  // uniform per warp
  if constexpr (ALIGNED) {
    if (inside)
      multi_tile2<K, FB, U, SEG, GUARDS, PF, 0>(a, mf, n, seg_active, f0, x0, ob, oe, lane, ring_base);
    else
      multi_tile2<K, FB, U, SEG, GUARDS, PF, 1>(a, mf, n, seg_active, f0, x0, ob, oe, lane, ring_base);
  } else {
    multi_tile2<K, FB, U, SEG, GUARDS, PF, 2>(a, mf, n, seg_active, f0, x0, ob, oe, lane, ring_base);
  }
}

}  // namespace c2d

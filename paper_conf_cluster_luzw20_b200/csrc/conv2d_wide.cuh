// conv2d_wide.cuh -- the single-channel kernel with 8 contiguous output columns per lane ("wide lanes").
//
// Same method as k_conv2d_single (conv2d_kernels.cuh): column reuse (Sec. II-A, Alg. 1
// the K-1 overlapping columns a lane needs beyond its own come from neighbouring lanes by
// warp shuffle, static register indices) and row reuse (Sec. II-B, Alg. 2: each input row
// is multiplied into K output-row accumulators held in registers). What changes is the lane's share:
//   * lane l owns the 8 CONTIGUOUS columns x0 + 8l .. x0 + 8l + 7 of a 256-column warp tile (the
//     one-warp-tile kernel: 4 contiguous columns per 128-column chunk, U chunks). The K-1 halo columns
//     are then K-1 shuffles (+ K-1 selects) per row for 8 outputs instead of per 4 -- the column-reuse
//     cost per output halves -- and one filter-row fetch (LDCU, uniform registers) feeds 8 columns;
//   * per input row a lane issues K*K*8 FFMA against ~(2K + K*ceil(K/4) + 20) other instructions:
//     94% FFMA at K = 15, 89% at K = 7 (the one-chunk kernel: 87% / 83%); the FMA-bound K >= 7 images
//     are issue-bound, so this is the lever.
// Halo element m (8 <= m < 8+K-1) of lane l is register m%8 of lane l + m/8; lanes 0 and 1 also hold
// the 16 columns right of the warp's span (the next tile's first two lanes), which the wrapping lanes
// 30/31 receive: the supplying lane selects (static index) its own register or its halo register --
// Alg. 1's select, generalised -- then one SHFL.IDX.
// Per output the terms are summed in filter-row, filter-column order (a FMA chain per output), the
// same order as the one-chunk kernel: the two kernels give the same bits, band- and batch-independent.
#pragma once

#include "conv2d_kernels.cuh"

namespace c2d {

constexpr int kWideV = 8;                 // contiguous output columns per lane
constexpr int kWideSpan = kWarp * kWideV;  // 256 columns per warp tile

template <int K>
struct WideCfg {
  static constexpr int WN = kWideV + K - 1;  // window per lane: 8 outputs + K-1 halo columns
  static constexpr int KP = (K + 3) / 4 * 4;
};

struct WideRow {
  float a[kWideV];  // own 8 columns
  float e[kWideV];  // lanes 0/1: the 8 columns at x0 + 256 + 8*lane (halo of lanes 31/30)
};

// a1: one input row of the tile. The warp is split into 32/SEG segments of SEG lanes (multi-channel:
// one image per segment; single-channel: SEG = 32); segment lane sl owns columns x0 + 8*sl .. + 7 and
// segment lanes 0/1 also hold the 16 columns right of the segment's span (x0 + 8*SEG + 8*sl).
// EDGE 0: 16B-aligned, every column of the span + halo inside the row: 2 x LDG.128 own + 2 x LDG.128
// halo (lanes >= 2 re-read lanes 0/1's halo: branch-free, same sectors). EDGE 1: aligned rows, ragged
// right edge: quad addresses clamped to the row's last quad (a valid output only reads inside quads;
// clamped garbage reaches only outputs >= Wo, never stored). EDGE 2: misaligned rows: guarded scalar
// loads.
template <int K, int EDGE, int SEG = kWarp>
__device__ __forceinline__ void wide_load(WideRow &b, const float *__restrict__ rowp, int x0, int Wc, int sl) {
  const int xa = x0 + kWideV * sl;
  const int xe = x0 + kWideV * SEG + kWideV * (sl & 1);
  if constexpr (EDGE == 2) {
#pragma unroll
    for (int t = 0; t < kWideV; ++t) b.a[t] = (xa + t < Wc) ? __ldg(rowp + xa + t) : 0.f;
#pragma unroll
    for (int t = 0; t < kWideV; ++t) b.e[t] = (K > 1 && xe + t < Wc) ? __ldg(rowp + xe + t) : 0.f;
  } else {
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int x = (EDGE == 1) ? min(xa + 4 * h, Wc - 4) : xa + 4 * h;
      const float4 v = ldg4(rowp + x);
      b.a[4 * h] = v.x; b.a[4 * h + 1] = v.y; b.a[4 * h + 2] = v.z; b.a[4 * h + 3] = v.w;
    }
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      if (K > 1 && 4 * h < K - 1) {  // static: only the halo quads the window uses
        const int x = (EDGE == 1) ? min(xe + 4 * h, Wc - 4) : xe + 4 * h;
        const float4 v = ldg4(rowp + x);
        b.e[4 * h] = v.x; b.e[4 * h + 1] = v.y; b.e[4 * h + 2] = v.z; b.e[4 * h + 3] = v.w;
      } else {
        b.e[4 * h] = b.e[4 * h + 1] = b.e[4 * h + 2] = b.e[4 * h + 3] = 0.f;
      }
    }
  }
}

// cp.async ring of wide rows: each lane copies its own 2 quads + its 2 halo quads global -> shared and
// later reads back only what it wrote (no cross-lane synchronisation), NST stages per warp.
template <int K, int NST, int SEG = kWarp>
struct WideRing {
  static constexpr unsigned kStageBytes = kWarp * 4 * 16;  // 4 quads per lane
  static constexpr unsigned kBytes = NST * kStageBytes;
  unsigned base;
  int lane, sl;
  __device__ __forceinline__ void issue(int stage, const float *__restrict__ rowp, int x0, int Wc, bool clamp) const {
    const unsigned sb = base + stage * kStageBytes + lane * 16;
    const int xa = x0 + kWideV * sl;
    const int xe = x0 + kWideV * SEG + kWideV * (sl & 1);
#pragma unroll
    for (int h = 0; h < 2; ++h) cp_async16(sb + h * kWarp * 16, rowp + (clamp ? min(xa + 4 * h, Wc - 4) : xa + 4 * h));
#pragma unroll
    for (int h = 0; h < 2; ++h)
      if (K > 1 && 4 * h < K - 1)
        cp_async16(sb + (2 + h) * kWarp * 16, rowp + (clamp ? min(xe + 4 * h, Wc - 4) : xe + 4 * h));
    cp_async_commit();
  }
  __device__ __forceinline__ void read(int stage, WideRow &b) const {
    const unsigned sb = base + stage * kStageBytes + lane * 16;
#pragma unroll
    for (int h = 0; h < 2; ++h) lds4_at(sb + h * kWarp * 16, b.a[4 * h], b.a[4 * h + 1], b.a[4 * h + 2], b.a[4 * h + 3]);
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      if (K > 1 && 4 * h < K - 1)
        lds4_at(sb + (2 + h) * kWarp * 16, b.e[4 * h], b.e[4 * h + 1], b.e[4 * h + 2], b.e[4 * h + 3]);
      else
        b.e[4 * h] = b.e[4 * h + 1] = b.e[4 * h + 2] = b.e[4 * h + 3] = 0.f;
    }
  }
};

// a2: w[0..WN) = in[x0 + 8*sl .. + WN). Halo element m (m >= 8) of segment lane sl is register m%8 of
// segment lane sl + m/8; a supplying lane s < m/8 serves a wrapped receiver (sl = s - m/8 + SEG) from
// its halo register. Shuffles stay inside the segment.
template <int K, int SEG = kWarp>
__device__ __forceinline__ void wide_window(const WideRow &b, float (&w)[WideCfg<K>::WN], int lane) {
  const int sl = lane & (SEG - 1);
  const int base = lane & ~(SEG - 1);
#pragma unroll
  for (int t = 0; t < kWideV; ++t) w[t] = b.a[t];
#pragma unroll
  for (int m = kWideV; m < WideCfg<K>::WN; ++m) {
    const int d = m / kWideV;  // source lane offset (static, 1 or 2)
    const int r = m % kWideV;  // source register (static)
    const float sup = (sl < d) ? b.e[r] : b.a[r];
    w[m] = __shfl_sync(kFull, sup, base | ((sl + d) & (SEG - 1)));
  }
}

// a4: filter rows of a KH x KW filter (rows padded to KP = ceil(KW/4)*4 floats): the per-K constant slot
// (uniform registers, square filters) or the CTA's shared-memory copy (broadcast LDS.128).
template <int KH, int KW, int FSRC>
struct FilterRows {
  static constexpr int KP = (KW + 3) / 4 * 4;
  unsigned sbase;
  const float *cbase;
  __device__ __forceinline__ void row(float (&fr)[KP], int i) const {
    if constexpr (FSRC == FSRC_CONST) {
      const float4 *p = reinterpret_cast<const float4 *>(cbase + i * KP);
#pragma unroll
      for (int c = 0; c < KP / 4; ++c) {
        const float4 v = p[c];
        fr[4 * c] = v.x; fr[4 * c + 1] = v.y; fr[4 * c + 2] = v.z; fr[4 * c + 3] = v.w;
      }
    } else {
#pragma unroll
      for (int c = 0; c < KP / 4; ++c)
        lds4_at(sbase + static_cast<unsigned>((i * KP + 4 * c) * 4), fr[4 * c], fr[4 * c + 1], fr[4 * c + 2],
                fr[4 * c + 3]);
    }
  }
};

// a3: one input row into the KH-slot ring: acc[q] = acc[q+1] + w . filter[KH-1-q] (shift folded into
// the FMA chains, static indices). GUARD: only slots qmin <= q < qmax (Alg. 2 cases 1 / 3, warp-uniform).
template <int KH, int KW, int FSRC, bool GUARD>
__device__ __forceinline__ void wide_step(float (&acc)[KH][kWideV], const float (&w)[WideCfg<KW>::WN],
                                          const FilterRows<KH, KW, FSRC> &fs, int qmin, int qmax) {
#pragma unroll
  for (int q = 0; q < KH; ++q) {
    if (!GUARD || (q >= qmin && q < qmax)) {
      float fr[FilterRows<KH, KW, FSRC>::KP];
      fs.row(fr, KH - 1 - q);
#pragma unroll
      for (int v = 0; v < kWideV; ++v) {
        float s = (q + 1 < KH) ? acc[(q + 1 < KH) ? q + 1 : 0][v] : 0.f;
#pragma unroll
        for (int j = 0; j < KW; ++j) s = fmaf(w[v + j], fr[j], s);
        acc[q][v] = s;
      }
    }
  }
}

// a6: the 8 outputs of every lane into a 256-column output chunk starting at g (16-byte alignment of g
// unknown: S = (g / 4) % 4 floats past a boundary, warp-uniform). S = 0: two STG.128 per lane. S > 0:
// lane l stores the aligned quads [8l+4-S, 8l+8-S) (own values) and [8l+8-S, 8l+12-S) (own o[8-S..7] +
// lane l+1's o[0..3-S], shfl.down); lane 0 the 4-S head columns, lane 31 its S tail columns (scalars).
template <int S>
__device__ __forceinline__ void wide_store_shifted(float *g, const float (&o)[kWideV], int lane) {
  if constexpr (S == 0) {
    stg4(g + kWideV * lane, o[0], o[1], o[2], o[3]);
    stg4(g + kWideV * lane + 4, o[4], o[5], o[6], o[7]);
  } else {
    float nb[4];
#pragma unroll
    for (int t = 0; t < 4; ++t) nb[t] = (t < 4 - S) ? __shfl_down_sync(kFull, o[t], 1) : 0.f;
    float* base = g + kWideV * lane;
    stg4(base + 4 - S, o[4 - S], o[5 - S], o[6 - S], o[7 - S]);
    float q[4];
#pragma unroll
    for (int k = 0; k < 4; ++k) q[k] = (k < S) ? o[(8 - S + k) & 7] : nb[(k - S) & 3];
    if (lane < kWarp - 1) stg4(base + 8 - S, q[0], q[1], q[2], q[3]);
    if (lane == 0) {
#pragma unroll
      for (int t = 0; t < 4 - S; ++t) __stcs(g + t, o[t]);
    }
    if (lane == kWarp - 1) {
#pragma unroll
      for (int t = 8 - S; t < 8; ++t) __stcs(base + t, o[t]);
    }
  }
}

template <bool SAFE>
__device__ __forceinline__ void wide_store(float *__restrict__ orow, int x0, int Wo, const float (&o)[kWideV],
                                           int lane) {
  if constexpr (!SAFE) {
    float *g = orow + x0;
    switch (static_cast<int>((reinterpret_cast<uintptr_t>(g) >> 2) & 3)) {  // warp-uniform
      case 0: wide_store_shifted<0>(g, o, lane); break;
      case 1: wide_store_shifted<1>(g, o, lane); break;
      case 2: wide_store_shifted<2>(g, o, lane); break;
      default: wide_store_shifted<3>(g, o, lane); break;
    }
  } else {
#pragma unroll
    for (int t = 0; t < kWideV; ++t) {
      const int x = x0 + kWideV * lane + t;
      if (x < Wo) __stcs(orow + x, o[t]);
    }
  }
}

// One warp tile: 256 columns x output rows [ob, oe), input rows [ob, oe+K-1) streamed once (Alg. 2's
// three cases as in single_tile). PF 1 / 2: the next one / two rows in flight in registers; PF >= 3
// (power of two, EDGE < 2): a PF-stage cp.async ring, PF-1 rows in flight. GUARDS as single_tile.
template <int KH, int KW, int FSRC, int PF, int GUARDS, int EDGE, bool HALO>
__device__ __forceinline__ void wide_tile(const SingleArgs &a, const float *__restrict__ inb, float *__restrict__ outb,
                                          const FilterRows<KH, KW, FSRC> &fs, int x0, int ob, int oe, int lane,
                                          unsigned ring_base) {
  constexpr bool SAFE = (EDGE != 0);
  constexpr int NST = (PF >= 3 && EDGE != 2) ? PF : 1;
  static_assert(NST == 1 || (NST & (NST - 1)) == 0, "ring depth must be a power of two");
  const int rend = oe + KH - 1;
  const int rlast = rend - 1;
  float acc[KH][kWideV];
#pragma unroll
  for (int q = 0; q < KH; ++q)
#pragma unroll
    for (int v = 0; v < kWideV; ++v) acc[q][v] = 0.f;
  WideRing<KW, (NST > 1 ? NST : 2)> ring;
  ring.base = ring_base;
  ring.lane = lane;
  ring.sl = lane;
  WideRow n1, n2;  // register path: rows r+1 (and r+2 when PF == 2) in flight
  if constexpr (NST > 1) {
#pragma unroll
    for (int st = 0; st < NST - 1; ++st) ring.issue(st, in_row<HALO>(a, inb, min(ob + st, rlast)), x0, a.Wc, EDGE == 1);
  } else {
    wide_load<KW, EDGE>(n1, in_row<HALO>(a, inb, ob), x0, a.Wc, lane);
    if constexpr (PF == 2) wide_load<KW, EDGE>(n2, in_row<HALO>(a, inb, min(ob + 1, rlast)), x0, a.Wc, lane);
  }
  // returns row r and issues the fetch of row r + depth (index clamped). PF == 2: the copy n1 = n2 reads
  // a row fetched one full iteration earlier, so it never waits on the load (PF == 1's cur = n1 copy
  // stalls on a load issued late in the previous iteration -- ncu long_scoreboard at that MOV).
  auto next_row = [&](int r) {
    WideRow cur;
    if constexpr (NST > 1) {
      cp_async_wait<NST - 2>();
      const int k = r - ob;
      ring.read(k & (NST - 1), cur);
      ring.issue((k + NST - 1) & (NST - 1), in_row<HALO>(a, inb, min(r + NST - 1, rlast)), x0, a.Wc, EDGE == 1);
    } else if constexpr (PF == 2) {
      cur = n1;
      n1 = n2;
      wide_load<KW, EDGE>(n2, in_row<HALO>(a, inb, min(r + 2, rlast)), x0, a.Wc, lane);
    } else {
      cur = n1;
      wide_load<KW, EDGE>(n1, in_row<HALO>(a, inb, min(r + 1, rlast)), x0, a.Wc, lane);
    }
    return cur;
  };
  auto out_at = [&](int o) { return outb + static_cast<size_t>(o) * a.Po; };
  int r = ob;
  if constexpr (GUARDS == 0) {
    for (; r < rend; ++r) {
      const WideRow cur = next_row(r);
      float w[WideCfg<KW>::WN];
      wide_window<KW>(cur, w, lane);
      wide_step<KH, KW, FSRC, false>(acc, w, fs, 0, KH);
      if (r >= ob + KH - 1) wide_store<SAFE>(out_at(r - KH + 1), x0, a.Wo, acc[0], lane);
    }
    return;
  }
  for (; r < min(ob + KH - 1, oe); ++r) {  // case 1: slots of outputs >= ob only
    const WideRow cur = next_row(r);
    float w[WideCfg<KW>::WN];
    wide_window<KW>(cur, w, lane);
    wide_step<KH, KW, FSRC, true>(acc, w, fs, KH - 1 - (r - ob), KH);
  }
  const int steady_end = (GUARDS == 2) ? oe : rend;
  for (; r < steady_end; ++r) {  // case 2 (+3 when GUARDS == 1)
    const WideRow cur = next_row(r);
    float w[WideCfg<KW>::WN];
    wide_window<KW>(cur, w, lane);
    wide_step<KH, KW, FSRC, false>(acc, w, fs, 0, KH);
    if (GUARDS == 2 || r >= ob + KH - 1) wide_store<SAFE>(out_at(r - KH + 1), x0, a.Wo, acc[0], lane);
  }
  for (; r < rend; ++r) {  // case 3 (GUARDS == 2): slots of outputs < oe only
    const WideRow cur = next_row(r);
    float w[WideCfg<KW>::WN];
    wide_window<KW>(cur, w, lane);
    wide_step<KH, KW, FSRC, true>(acc, w, fs, max(0, KH - 1 - (r - ob)), oe + KH - 1 - r);
    if (r >= ob + KH - 1) wide_store<SAFE>(out_at(r - KH + 1), x0, a.Wo, acc[0], lane);
  }
}

// One warp per CTA (warp-uniform control flow: the constant-slot filter stays in uniform registers).
// SingleArgs.n_cb counts 256-column blocks. KH x KW filter (square: KH = KW = K; rectangular filters,
// conv2d_single_rect, take the shared-memory filter).
// Rectangular instantiations state 8 resident CTAs (a 255-register cap): without it ptxas caps some
// (KH, KW) at 168 registers and spills (tests/test_sass.py); square ones keep ptxas' own choice unless
// MINB > 1 states the resident CTAs the register allocation must allow.
template <int KH, int KW, int FSRC, int PF, int GUARDS, bool HALO, int MINB = 1>
__global__ void __launch_bounds__(kWarp, (KH != KW) ? 8 : MINB) k_conv2d_wide(const SingleArgs a) {
  using FR = FilterRows<KH, KW, FSRC>;
  __shared__ __align__(16) float sf[(FSRC == FSRC_SMEM) ? KH * FR::KP : 4];
  extern __shared__ __align__(16) float wide_ring_smem[];
  FR fs;
  if constexpr (FSRC == FSRC_CONST) {
    fs.cbase = c_filt;
  } else {
    for (int t = threadIdx.x; t < KH * FR::KP; t += blockDim.x) {
      const int i = t / FR::KP, j = t % FR::KP;
      sf[t] = (j < KW) ? a.filt[i * KW + j] : 0.f;
    }
    __syncwarp();
    fs.sbase = static_cast<unsigned>(__cvta_generic_to_shared(sf));
  }
  const int lane = threadIdx.x;
  const int tile = static_cast<int>(blockIdx.x);
  const unsigned ring_base = static_cast<unsigned>(__cvta_generic_to_shared(wide_ring_smem));
  const int cb = tile % a.n_cb;
  const int t2 = tile / a.n_cb;
  const int band = t2 % a.n_bands;
  const int img = t2 / a.n_bands;
  const float *__restrict__ inb = a.in + img * a.img_in;
  float *__restrict__ outb = a.out + img * a.img_out;
  const int x0 = cb * kWideSpan;
  const int ob = band_start(band, a.n_bands, a.Ho);
  const int oe = band_start(band + 1, a.n_bands, a.Ho);
  const bool inside = x0 + kWideSpan + 16 <= a.W;  // span + both halo quads in range (warp-uniform)
  if (a.aligned && inside)
    wide_tile<KH, KW, FSRC, PF, GUARDS, 0, HALO>(a, inb, outb, fs, x0, ob, oe, lane, ring_base);
  else if (a.aligned)
    wide_tile<KH, KW, FSRC, PF, GUARDS, 1, HALO>(a, inb, outb, fs, x0, ob, oe, lane, ring_base);
  else
    wide_tile<KH, KW, FSRC, PF, GUARDS, 2, HALO>(a, inb, outb, fs, x0, ob, oe, lane, ring_base);
}

}  // namespace c2d

// conv2d_pair.cuh -- the one-chunk single-channel kernel with its row-reuse ring run as PAIRED FMAs.
//
// Row reuse (Sec. II-B, Alg. 2) keeps K output-row accumulators per column, slot q
// holding output row r-K+1+q after input row r; each input row adds w . filter[K-1-q] to slot q (and
// shifts the ring). The one-chunk kernel (k_conv2d_single, U = 1) does this with 15x15x4 = 900 scalar
// FFMA per row at K = 15 and is issue-bound (ncu: issue 93%, FMA pipe 80%, 14% of the issued
// instructions are the shuffles, filter fetches, loads, stores and loop control).
//
// sm_100's FFMA2 (fma.rn.f32x2) runs two FMA chains in one instruction, with a scalar-broadcast register
// operand and a uniform-register PAIR operand. Here it pairs two ring slots of the same column: for odd
// K, H = (K+1)/2, slot q and slot q+H (q = 0..H-2) share the window value w[v+j] (the broadcast) and
// read the filter pair (f[K-1-q][j], f[K-1-q-H][j]) as one UR pair. The ring shift keeps the pairing:
// pair q takes pair q+1's values. The middle slot H-1 has no partner: it runs as a scalar chain (its
// input is pair 0's upper half, slot H), and is kept as a register pair with a zero upper half, so the
// last pair (H-2, K-1) reads it as (slot H-1, 0) -- the shift-in of a fresh slot K-1 -- without a copy.
// Per row at K = 15: 7 pairs x 4 columns x 15 taps = 420 FFMA2 + 60 FFMA for the 900 FMAs, about 630
// issue slots against 900 FMA-pipe cycles: the FMA pipe, not the issue port, becomes the bound.
// Each output still sums filter rows ascending, taps ascending, one round-to-nearest FMA each: the same
// bits as the scalar kernels (band-, batch- and row-band independent).
//
// The filter lives in the unit's constant slot as a pair table (tools/..., launch.cuh: three
// stream-ordered copies, two of them interleaving 4-byte elements at an 8-byte pitch):
//   pairs  [p][j] = (f[H+p][j], f[p][j])   p = 0..H-2 (pair p serves ring slots H-2-p and K-2-p)
//   single [j]    =  f[H-1][j]             at float offset kPairSingle
#pragma once

#include "conv2d_kernels.cuh"

namespace c2d {

template <int K>
struct PairCfg {
  static_assert(K % 2 == 1 && K >= 3, "odd K");
  static constexpr int H = (K + 1) / 2;
  static constexpr int NP = H - 1;                              // slot pairs
  static constexpr int kSingle = (NP * K * 2 + 3) / 4 * 4;    // float offset of the single row
  static constexpr int kFloats = kSingle + (K + 3) / 4 * 4;
  static_assert(kFloats <= kConstSlotFloats, "constant slot");
};

// One input row into the paired ring (U = 1: 4 columns per lane). P[q][v] = (slot q, slot q+H) of column
// v, S[v] = (slot H-1, 0).
template <int K>
__device__ __forceinline__ void pair_step(float2 (&P)[PairCfg<K>::NP][4], float2 (&S)[4],
                                          const float (&w)[KCfg<K>::WN], const float *cbase) {
  constexpr int H = PairCfg<K>::H, NP = PairCfg<K>::NP;
  const float2 *pt = reinterpret_cast<const float2 *>(cbase);
  const float *st = cbase + PairCfg<K>::kSingle;
  float2 nS[4];
  // the middle slot: S' = slot H (pair 0's upper half) + w . f[H-1]
#pragma unroll
  for (int v = 0; v < 4; ++v) {
    float s = P[0][v].y;
#pragma unroll
    for (int j = 0; j < K; ++j) s = fmaf(w[v + j], st[j], s);
    nS[v] = make_float2(s, 0.f);
  }
  // pairs q = 0..H-2: P'(q) = P(q+1) (P(H-2): S) + w . (f[K-1-q], f[K-1-q-H]); table row p = H-2-q
#pragma unroll
  for (int q = 0; q < NP; ++q) {
    const int p = NP - 1 - q;
#pragma unroll
    for (int v = 0; v < 4; ++v) {
      float2 s = (q + 1 < NP) ? P[(q + 1 < NP) ? q + 1 : 0][v] : S[v];
#pragma unroll
      for (int j = 0; j < K; ++j) s = __ffma2_rn(make_float2(w[v + j], w[v + j]), pt[p * K + j], s);
      P[q][v] = s;
    }
  }
#pragma unroll
  for (int v = 0; v < 4; ++v) S[v] = nS[v];
}

// One warp tile (U = 1, 128 columns) x output rows [ob, oe), every row through the full paired ring
// (Alg. 2 cases 1 and 3 unguarded: their extra FMAs land in slots that are never stored). Row fetch as
// single_tile: PF 1 (next row in registers) or a PF-stage cp.async ring.
template <int K, int PF, int EDGE, bool HALO>
__device__ __forceinline__ void pair_tile(const SingleArgs &a, const float *__restrict__ inb, float *__restrict__ outb,
                                          int x0, int ob, int oe, int lane, unsigned ring_base) {
  constexpr int NP = PairCfg<K>::NP;
  constexpr bool SAFE = (EDGE != 0);
  constexpr int NST = (PF >= 3 && EDGE != 2) ? PF : 1;
  const int rend = oe + K - 1;
  const int rlast = rend - 1;
  float2 P[NP][4], S[4];
#pragma unroll
  for (int q = 0; q < NP; ++q)
#pragma unroll
    for (int v = 0; v < 4; ++v) P[q][v] = make_float2(0.f, 0.f);
#pragma unroll
  for (int v = 0; v < 4; ++v) S[v] = make_float2(0.f, 0.f);
  RowRing<K, 1, kWarp, (NST > 1 ? NST : 2)> ring;
  ring.base = ring_base;
  ring.lane = lane;
  ring.sl = lane;
  constexpr bool clamp = (EDGE == 1);
  RowBuf<K, 1> n1;
  if constexpr (NST > 1) {
#pragma unroll
    for (int st = 0; st < NST - 1; ++st) ring.issue(st, in_row<HALO>(a, inb, min(ob + st, rlast)), x0, a.Wc, clamp);
  } else {
    load_row<K, 1, SAFE>(n1, in_row<HALO>(a, inb, ob), x0, a.Wc, lane, a.aligned);
  }
  for (int r = ob; r < rend; ++r) {
    RowBuf<K, 1> cur;
    if constexpr (NST > 1) {
      cp_async_wait<NST - 2>();
      const int k = r - ob;
      ring.read(k & (NST - 1), cur);
      ring.issue((k + NST - 1) & (NST - 1), in_row<HALO>(a, inb, min(r + NST - 1, rlast)), x0, a.Wc, clamp);
    } else {
      cur = n1;
      load_row<K, 1, SAFE>(n1, in_row<HALO>(a, inb, min(r + 1, rlast)), x0, a.Wc, lane, a.aligned);
    }
    float w[1][KCfg<K>::WN];
    build_windows<K, 1>(cur, w, lane);
    pair_step<K>(P, S, w[0], c_filt);
    if (r >= ob + K - 1) {
      float o[1][4];
#pragma unroll
      for (int v = 0; v < 4; ++v) o[0][v] = P[0][v].x;  // slot 0: output row r-K+1, complete
      store_row<1, SAFE>(outb + static_cast<size_t>(r - K + 1) * a.Po, x0, a.Wo, o, lane);
    }
  }
}

// One warp per CTA (warp-uniform control flow: the pair table stays in uniform registers).
template <int K, int PF, bool HALO>
__global__ void __launch_bounds__(kWarp) k_conv2d_pair(const SingleArgs a) {
  extern __shared__ __align__(16) float pair_ring_smem[];
  const int lane = threadIdx.x;
  const int tile = static_cast<int>(blockIdx.x);
  const unsigned ring_base = static_cast<unsigned>(__cvta_generic_to_shared(pair_ring_smem));
  const int cb = tile % a.n_cb;
  const int t2 = tile / a.n_cb;
  const int band = t2 % a.n_bands;
  const int img = t2 / a.n_bands;
  const float *__restrict__ inb = a.in + img * a.img_in;
  float *__restrict__ outb = a.out + img * a.img_out;
  const int x0 = cb * 128;
  const int ob = band_start(band, a.n_bands, a.Ho);
  const int oe = band_start(band + 1, a.n_bands, a.Ho);
  const bool inside = x0 + 128 + 4 * KCfg<K>::NE <= a.W;
  if (a.aligned && inside)
    pair_tile<K, PF, 0, HALO>(a, inb, outb, x0, ob, oe, lane, ring_base);
  else if (a.aligned)
    pair_tile<K, PF, 1, HALO>(a, inb, outb, x0, ob, oe, lane, ring_base);
  else
    pair_tile<K, PF, 2, HALO>(a, inb, outb, x0, ob, oe, lane, ring_base);
}

}  // namespace c2d

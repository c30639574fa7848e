// conv2d_split.cuh -- single-channel kernel with the filter rows split across a thread-block cluster.
//
// Row reuse (Sec. II-B, Alg. 2) streams the IH = BH + K - 1 input rows of a band
// through a K-slot ring; the first K-1 of them (Alg. 2 case 1) complete no output, so a band of BH
// output rows pays (BH + K - 1) / BH row fetches, shuffles and ring steps per output row. On B200 the
// band height is not free: a full wave of warps over a 1K-4K image leaves BH of 4-60 rows, and the
// case-1 rows then cost up to several times the useful work (K = 15: 14 extra rows per band).
//
// This kernel runs one warp tile (128*U columns x BH output rows) on a CLUSTER of G one-warp CTAs.
// CTA g of the cluster owns filter rows [g*K/G, (g+1)*K/G) -- KG of them -- and applies Alg. 2 to
// those rows only: it streams input rows [ob + I0, oe + I0 + KG - 1) through a KG-slot ring, so its
// case-1 prologue is KG - 1 rows instead of K - 1, and each CTA's ring (and register file) is KG/K
// of the full one. The G partial output rows are summed through distributed shared memory:
//   * every CTA writes its partial rows into its own shared memory, R rows per chunk, 3 chunk
//     buffers (triple buffering: chunk c+1 is computed while chunk c is being reduced);
//   * after a cluster barrier (one per chunk; release / acquire fences restricted to shared memory), CTA g
//     reduces the rows k = g, g+G, ... of the chunk: it reads the G partials of each row from the G
//     CTAs' shared memory (ld.shared::cluster via mapa), adds them in rank order 0..G-1, and stores
//     the output row (a6, the same coalesced / realigned store as the one-CTA kernel);
//   * the barrier of chunk c+1 also certifies that every CTA finished reading chunk c-1, so the
//     buffer of chunk c+2 (= c-1 mod 3) is free when it is written.
// Per output the terms are summed as: within a CTA filter rows ascending (each in column order), then
// the G partials in rank order -- a fixed order that depends on (K, G) only, not on the band, so
// outputs are band-position independent (row-band sharding stays bitwise).
// The filter comes from the per-K constant slot (uniform registers): every CTA is one warp and every
// branch depends on blockIdx, the cluster rank and kernel parameters only.
#pragma once

#include "conv2d_kernels.cuh"

namespace c2d {

struct SplitArgs {
  const float *in;
  const float *in2;  // rows >= H1 at in2 (row-band halo), as SingleArgs
  int H1;
  int P;        // input row pitch in floats, as SingleArgs
  int Wc;       // row-fetch bound, as SingleArgs
  int Po;       // output row pitch, as SingleArgs
  float *out;
  int H, W, Ho, Wo;
  int n_img;          // images of a batch, as SingleArgs
  long long img_in;   // floats between consecutive input images
  long long img_out;  // floats between consecutive output images
  int n_bands;  // balanced output-row bands per image (band_start)
  int n_cb;     // column blocks of 128*U outputs
  int n_tiles;  // n_img * n_bands * n_cb (clusters)
  int aligned;  // in is 16B aligned and W % 4 == 0
};

__device__ __forceinline__ unsigned cluster_ctarank() {
  unsigned r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
  return r;
}
// Arrive with release semantics restricted to this CTA's shared-memory writes (the partial rows):
// MEMBAR.ALL.CTA instead of the MEMBAR.ALL.GPU of barrier.cluster.arrive.release, which would also
// wait for this warp's outstanding global output stores and row prefetches.
__device__ __forceinline__ void cluster_arrive() {
  asm volatile("fence.release.sync_restrict::shared::cta.cluster;" ::: "memory");
  asm volatile("barrier.cluster.arrive.relaxed.aligned;" ::: "memory");
}
__device__ __forceinline__ void cluster_wait() {
  asm volatile("barrier.cluster.wait.aligned;" ::: "memory");
  asm volatile("fence.acquire.sync_restrict::shared::cluster.cluster;" ::: "memory");
}
// shared-window address of the same variable in CTA `rank` of the cluster
__device__ __forceinline__ unsigned mapa_rank(unsigned saddr, unsigned rank) {
  unsigned r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(saddr), "r"(rank));
  return r;
}
__device__ __forceinline__ float4 ld_dsmem4(unsigned caddr) {
  float4 v;
  asm volatile("ld.shared::cluster.v4.f32 {%0, %1, %2, %3}, [%4];"
               : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w)
               : "r"(caddr)
               : "memory");
  return v;
}
__device__ __forceinline__ void st_smem4(unsigned saddr, float a, float b, float c, float d) {
  asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(saddr), "f"(a), "f"(b), "f"(c), "f"(d) : "memory");
}

// Filter rows of cluster rank RANK: [I0, I0 + KG)
template <int K, int G, int RANK>
struct SplitRows {
  static constexpr int I0 = RANK * K / G;
  static constexpr int KG = (RANK + 1) * K / G - I0;
};

// one input row into the KG-slot ring of filter rows I0..I0+KG-1: acc[q] = acc[q+1] + w . f[I0+KG-1-q]
// GUARD: only slots q >= qmin (the first KG-1 rows of a band feed only outputs >= ob)
template <int K, int KG, int I0, int U, bool GUARD>
__device__ __forceinline__ void row_step_split(float (&acc)[KG][U][4], const float (&w)[U][KCfg<K>::WN],
                                               const FilterSrc<K, FSRC_CONST> &fs, int qmin) {
#pragma unroll
  for (int q = 0; q < KG; ++q) {
    if (!GUARD || q >= qmin) {
      float fr[KCfg<K>::KP];
      fs.row(fr, I0 + KG - 1 - q);
#pragma unroll
      for (int u = 0; u < U; ++u) {
#pragma unroll
        for (int v = 0; v < 4; ++v) {
          float s = (q + 1 < KG) ? acc[(q + 1 < KG) ? q + 1 : 0][u][v] : 0.f;
#pragma unroll
          for (int j = 0; j < K; ++j) s = fmaf(w[u][v + j], fr[j], s);
          acc[q][u][v] = s;
        }
      }
    }
  }
}

template <int U, int R>
struct SplitBuf {
  static constexpr unsigned kRowBytes = U * kWarp * 16;  // one partial row: U float4 per lane
  static constexpr unsigned kChunkBytes = R * kRowBytes;
  static constexpr unsigned kBytes = 3 * kChunkBytes;
};

// One cluster tile, this CTA's share: filter rows of rank RANK, outputs [ob, oe), columns x0.
// CL = 1: the G parts are the one-warp CTAs of a cluster (partials read through DSMEM, cluster
// barriers); CL = 0: the G parts are the G warps of one CTA (partials in the CTA's shared memory,
// named barrier). smem0: this CTA's dynamic shared memory; each part owns PW bytes of it (CL = 0: at
// RANK * PW) holding its 3 chunk buffers and its row ring.
template <int K, int G, int RANK, int U, int PF, int R, int GUARDS, int EDGE, int CL>
__device__ __forceinline__ void split_tile(const SplitArgs &a, const float *__restrict__ inb,
                                           float *__restrict__ outb, const FilterSrc<K, FSRC_CONST> &fs, int x0,
                                           int ob, int oe, int lane, unsigned smem0, unsigned PW) {
  constexpr int I0 = SplitRows<K, G, RANK>::I0;
  constexpr int KG = SplitRows<K, G, RANK>::KG;
  constexpr bool SAFE = (EDGE != 0);
  constexpr int NST = (PF >= 3 && EDGE != 2) ? PF : 1;
  static_assert(NST == 1 || (NST & (NST - 1)) == 0, "ring depth must be a power of two");
  using Buf = SplitBuf<U, R>;
  const unsigned buf_base = smem0 + (CL ? 0u : RANK * PW);
  const unsigned ring_base = buf_base + Buf::kBytes;
  // partial row k of chunk buffer cb_off, part g
  auto part_addr = [&](unsigned off, int g) -> unsigned {
    if constexpr (CL) return mapa_rank(smem0 + off, g);
    else return smem0 + g * PW + off;
  };
  auto part_ld = [&](unsigned addr) -> float4 {
    if constexpr (CL) {
      return ld_dsmem4(addr);
    } else {
      float4 v;
      lds4_at(addr, v.x, v.y, v.z, v.w);
      return v;
    }
  };
  auto sync_wait = [&]() {
    if constexpr (CL) cluster_wait();
    else asm volatile("bar.sync 1, %0;" ::"n"(G * kWarp) : "memory");
  };
  auto sync_arrive = [&]() {
    if constexpr (CL) cluster_arrive();
  };
  const int r0 = ob + I0;            // first input row of this CTA
  const int rend = oe + I0 + KG - 1;  // input rows [r0, rend)
  const int rlast = rend - 1;
  float acc[KG][U][4];
#pragma unroll
  for (int q = 0; q < KG; ++q)
#pragma unroll
    for (int u = 0; u < U; ++u)
#pragma unroll
      for (int v = 0; v < 4; ++v) acc[q][u][v] = 0.f;
  RowRing<K, U, kWarp, (NST > 1 ? NST : 2)> ring;
  ring.base = ring_base;
  ring.lane = lane;
  ring.sl = lane;
  constexpr bool clamp = (EDGE == 1);
  RowBuf<K, U> n1;
  auto in_row_p = [&](int r) {
    return r < a.H1 ? inb + static_cast<size_t>(r) * a.P : a.in2 + static_cast<size_t>(r - a.H1) * a.P;
  };
  if constexpr (NST > 1) {
#pragma unroll
    for (int st = 0; st < NST - 1; ++st) ring.issue(st, in_row_p(min(r0 + st, rlast)), x0, a.Wc, clamp);
  } else {
    load_row<K, U, SAFE>(n1, in_row_p(r0), x0, a.Wc, lane, a.aligned);
  }
  int r = r0;
  auto next_row = [&]() {
    RowBuf<K, U> cur;
    if constexpr (NST > 1) {
      cp_async_wait<NST - 2>();
      const int k = r - r0;
      ring.read(k & (NST - 1), cur);
      ring.issue((k + NST - 1) & (NST - 1), in_row_p(min(r + NST - 1, rlast)), x0, a.Wc, clamp);
    } else {
      cur = n1;
      load_row<K, U, SAFE>(n1, in_row_p(min(r + 1, rlast)), x0, a.Wc, lane, a.aligned);
    }
    return cur;
  };
  // Alg. 2 case 1 on this CTA's rows: the first KG-1 input rows complete no output
  for (; r < min(r0 + KG - 1, rend); ++r) {
    const RowBuf<K, U> cur = next_row();
    float w[U][KCfg<K>::WN];
    build_windows<K, U>(cur, w, lane);
    if constexpr (GUARDS != 0)
      row_step_split<K, KG, I0, U, true>(acc, w, fs, KG - 1 - (r - r0));
    else
      row_step_split<K, KG, I0, U, false>(acc, w, fs, 0);
  }
  // reduce chunk c: rows k = RANK, RANK+G, ... of the chunk, partials of ranks 0..G-1 in order
  auto reduce_chunk = [&](int c, int rows_c) {
    const unsigned coff = (c % 3) * Buf::kChunkBytes;
    for (int k = RANK; k < rows_c; k += G) {
      float o[U][4];
#pragma unroll
      for (int g = 0; g < G; ++g) {
        const unsigned remote = part_addr(coff + k * Buf::kRowBytes, g);
#pragma unroll
        for (int u = 0; u < U; ++u) {
          const float4 p = part_ld(remote + (u * kWarp + lane) * 16);
          if (g == 0) {
            o[u][0] = p.x; o[u][1] = p.y; o[u][2] = p.z; o[u][3] = p.w;
          } else {
            o[u][0] += p.x; o[u][1] += p.y; o[u][2] += p.z; o[u][3] += p.w;
          }
        }
      }
      float *orow = outb + static_cast<size_t>(ob + c * R + k) * a.Po;
      store_row<U, SAFE>(orow, x0, a.Wo, o, lane);
    }
  };
  // Alg. 2 case 2 (+3): one output row per input row, R per chunk
  const int n_out = oe - ob;
  const int n_chunks = (n_out + R - 1) / R;
  for (int c = 0; c < n_chunks; ++c) {
    const int rows_c = min(R, n_out - c * R);
    const unsigned cb = buf_base + (c % 3) * Buf::kChunkBytes;
    for (int k = 0; k < rows_c; ++k, ++r) {
      const RowBuf<K, U> cur = next_row();
      float w[U][KCfg<K>::WN];
      build_windows<K, U>(cur, w, lane);
      row_step_split<K, KG, I0, U, false>(acc, w, fs, 0);
#pragma unroll
      for (int u = 0; u < U; ++u)
        st_smem4(cb + k * Buf::kRowBytes + (u * kWarp + lane) * 16, acc[0][u][0], acc[0][u][1], acc[0][u][2],
                 acc[0][u][3]);
    }
    if (c > 0) {
      sync_wait();  // chunk c-1 written by every part
      reduce_chunk(c - 1, R);
    }
    sync_arrive();  // chunk c written, chunk c-1 read
  }
  sync_wait();
  reduce_chunk(n_chunks - 1, n_out - (n_chunks - 1) * R);
  if constexpr (CL) {  // keep this CTA's shared memory alive until every CTA finished reading it
    cluster_arrive();
    cluster_wait();
  }
}

template <int K, int G, int U, int PF, int R, int GUARDS, int EDGE, int CL, int RK = 0>
__device__ __forceinline__ void split_dispatch(unsigned rank, const SplitArgs &a, const float *__restrict__ inb,
                                               float *__restrict__ outb, const FilterSrc<K, FSRC_CONST> &fs,
                                               int x0, int ob, int oe, int lane, unsigned smem0, unsigned PW) {
  if constexpr (RK < G) {
    if (rank == RK)
      split_tile<K, G, RK, U, PF, R, GUARDS, EDGE, CL>(a, inb, outb, fs, x0, ob, oe, lane, smem0, PW);
    else
      split_dispatch<K, G, U, PF, R, GUARDS, EDGE, CL, RK + 1>(rank, a, inb, outb, fs, x0, ob, oe, lane, smem0, PW);
  }
}

template <int K, int U, int PF, int R>
struct SplitSmem {  // bytes per part: 3 chunk buffers + the row ring
  static constexpr unsigned kPart =
      SplitBuf<U, R>::kBytes + ((PF >= 3) ? RowRing<K, U, kWarp, (PF >= 3 ? PF : 2)>::kBytes : 0u);
};

// CL = 1: grid n_tiles * G one-warp CTAs, cluster (G, 1, 1); CL = 0: grid n_tiles CTAs of G warps.
template <int K, int G, int U, int PF, int R, int GUARDS, int CL>
__global__ void __launch_bounds__(CL ? kWarp : G * kWarp) k_conv2d_split(const SplitArgs a) {
  extern __shared__ __align__(16) float split_smem[];
  FilterSrc<K, FSRC_CONST> fs;
  fs.cbase = c_filt;
  const int lane = threadIdx.x & (kWarp - 1);
  const unsigned rank = CL ? cluster_ctarank() : (threadIdx.x >> 5);
  const int tile = CL ? static_cast<int>(blockIdx.x) / G : static_cast<int>(blockIdx.x);
  const unsigned smem0 = static_cast<unsigned>(__cvta_generic_to_shared(split_smem));
  constexpr unsigned PW = SplitSmem<K, U, PF, R>::kPart;
  const int cb = tile % a.n_cb;
  const int t2 = tile / a.n_cb;
  const int band = t2 % a.n_bands;
  const int img = t2 / a.n_bands;
  const float *__restrict__ inb = a.in + img * a.img_in;
  float *__restrict__ outb = a.out + img * a.img_out;
  const int x0 = cb * 128 * U;
  const int ob = band_start(band, a.n_bands, a.Ho);
  const int oe = band_start(band + 1, a.n_bands, a.Ho);
  const bool inside = x0 + 128 * U + 4 * KCfg<K>::NE <= a.W;  // uniform over the cluster
  if (a.aligned && inside)
    split_dispatch<K, G, U, PF, R, GUARDS, 0, CL>(rank, a, inb, outb, fs, x0, ob, oe, lane, smem0, PW);
  else if (a.aligned)
    split_dispatch<K, G, U, PF, R, GUARDS, 1, CL>(rank, a, inb, outb, fs, x0, ob, oe, lane, smem0, PW);
  else
    split_dispatch<K, G, U, PF, R, GUARDS, 2, CL>(rank, a, inb, outb, fs, x0, ob, oe, lane, smem0, PW);
}

}  // namespace c2d

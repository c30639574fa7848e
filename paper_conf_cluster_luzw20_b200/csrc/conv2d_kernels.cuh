// conv2d_kernels.cuh -- sm_100a kernels for direct, stride-1, valid-mode fp32 convolution with the
// column reuse and row reuse of Lu, Zhang & Wang (Cluster 2020), re-designed for B200.
//
// Work decomposition:
//   * One WARP owns a tile of 128*U output columns x BH output rows ("band"). Lane l holds the
//     outputs x0 + 128u + 4l + {0..3} of every chunk u < U (V = 4 contiguous columns per lane, so
//     every input-row load is one coalesced LDG.128 per lane and every output store is STG.128).
//   * a1 Input row fetch: per input row, U LDG.128 per lane plus one extra LDG.128 for the K-1 halo
//     columns right of the warp's span (lanes >= NE = ceil((K-1)/4) re-read a duplicate quad so the
//     load is branch-free). The next row is in flight while the current one is computed.
//   * a2 Column reuse (Sec. II-A, Alg. 1, Fig. 1c): the K-1 halo values
//     a lane needs beyond its own 4 come from lanes l+1.. via __shfl_sync, never from memory. As in
//     Alg. 1, the value a lane SUPPLIES is chosen with a static register index and a lane-dependent
//     select (Alg. 1 lines 2-5 select by a 64-bit shift; here a SEL), so the window iTemp stays in
//     registers. Halo element m (m = 4..K+2) of lane l lives in register
//     m%4 of lane l + m/4: one SEL + one SHFL.IDX per (m, chunk), all indices compile-time.
//   * a3 Row reuse (Sec. II-B, Alg. 2, flow P:303-311): each loaded input row is
//     multiplied against all K filter rows into K output-row accumulators held in registers
//     ("out ... can be stored in registers"). Slot q of the ring holds output row
//     r-K+1+q after input row r; the update acc[q] = acc[q+1] + row . filter[K-1-q] SHIFTS the ring
//     inside the first FMA of each chain, so the ring rotation costs no MOVs and every index is
//     static (the dynamic->static index transformation of P:75-77). The first K-1 rows
//     of a band (Alg. 2 case 1) skip the slots whose output row precedes the band; Alg. 2 case 3 is
//     implicit (the band stops when its last output row completes).
//   * a4 Filter supply: a per-launch slot of the __constant__ bank read through uniform registers
//     (LDCU.128 + FFMA with a UR operand: one fetch serves the whole warp, no per-lane traffic), or
//     shared memory (broadcast LDS.128) when the launch is being captured into a CUDA graph.
//   * a5 Channel reduction (multi): for each input row, all C channels stream through the same
//     accumulators; each thread also carries FB filters, so one window feeds FB*K*K*4 FMAs.
//   * a6 Output store: slot 0 is complete after each row -> one coalesced store per lane; rows whose
//     pitch breaks 16-byte alignment are realigned with warp shuffles (static per-shift variants).
// Edge tiles (ragged right edge: clamped vector loads, masked stores) and misaligned tensors (scalar
// loads/stores) take the same code with SAFE=true.
#pragma once

#include <cstdint>
#include <cuda_runtime.h>

namespace c2d {

constexpr unsigned kFull = 0xffffffffu;
constexpr int kWarp = 32;
constexpr int kCtaWarps = 4;  // 128 threads per CTA

template <int K>
struct KCfg {
  static constexpr int NE = (K - 1 + 3) / 4;  // lanes that fetch the extra halo float4
  static constexpr int KP = (K + 3) / 4 * 4;  // filter row padded to a multiple of 4 floats
  static constexpr int WN = 4 + K - 1;        // window length per chunk: 4 outputs + K-1 halo
};

// ------------------------------------------------------------------------------------------------
// memory helpers
// ------------------------------------------------------------------------------------------------
__device__ __forceinline__ float4 ldg4(const float *p) { return __ldg(reinterpret_cast<const float4 *>(p)); }

__device__ __forceinline__ void stg4(float *p, float a, float b, float c, float d) {
  __stcs(reinterpret_cast<float4 *>(p), make_float4(a, b, c, d));
}

__device__ __forceinline__ void lds4_at(unsigned saddr, float &a, float &b, float &c, float &d) {
  asm volatile("ld.shared.v4.f32 {%0, %1, %2, %3}, [%4];" : "=f"(a), "=f"(b), "=f"(c), "=f"(d) : "r"(saddr));
}

// LDS.128 that the compiler may not hoist out of the row loop (keeps the staged filters out of the
// register file).
__device__ __forceinline__ void lds4_volatile(const float *p, float &a, float &b, float &c, float &d) {
  const unsigned s = static_cast<unsigned>(__cvta_generic_to_shared(p));
  asm volatile("ld.shared.v4.f32 {%0, %1, %2, %3}, [%4];" : "=f"(a), "=f"(b), "=f"(c), "=f"(d) : "r"(s));
}

// ------------------------------------------------------------------------------------------------
// a1: one input row segment of a warp tile
// ------------------------------------------------------------------------------------------------
template <int K, int U>
struct RowBuf {
  float a[U][4];
  float e[4];
};

// One row segment of a warp tile. The warp is split into 32/SEG segments of SEG lanes; segment lane
// sl holds columns x0 + 4*SEG*u + 4*sl + {0..3} of chunk u < U, plus (lanes sl < NE) one quad of the
// K-1 halo columns right of the segment's span. rowp points at input column 0 of the row.
//   SAFE == false: the whole span + halo is inside the row and 16-byte aligned: LDG.128 per lane,
//                  and every lane loads a halo quad (lanes >= NE re-read a duplicate: branch-free).
//   SAFE == true : ragged right edge or misaligned rows. Aligned rows (W % 4 == 0, 16-byte base):
//                  the quad address is clamped to the last quad of the row -- quads are either fully
//                  inside or fully outside the row, and a valid output only reads inside quads, so
//                  the clamped (garbage) values only reach outputs >= Wo, which are never stored.
//                  Misaligned rows: guarded scalar loads.
template <int K, int U, int SEG, bool SAFE>
__device__ __forceinline__ void load_row_g(RowBuf<K, U> &b, const float *__restrict__ rowp, int x0, int W, int sl,
                                           bool aligned) {
  constexpr int NE = KCfg<K>::NE;
#pragma unroll
  for (int u = 0; u < U; ++u) {
    const int x = x0 + 4 * SEG * u + 4 * sl;
    if (!SAFE || aligned) {
      const float4 v = ldg4(rowp + (SAFE ? min(x, W - 4) : x));
      b.a[u][0] = v.x; b.a[u][1] = v.y; b.a[u][2] = v.z; b.a[u][3] = v.w;
    } else {
#pragma unroll
      for (int t = 0; t < 4; ++t) b.a[u][t] = (x + t < W) ? __ldg(rowp + x + t) : 0.f;
    }
  }
  const int xe = x0 + 4 * SEG * U + 4 * (sl % (NE > 0 ? NE : 1));
  if constexpr (NE == 0) {
#pragma unroll
    for (int t = 0; t < 4; ++t) b.e[t] = 0.f;
  } else {
    if (!SAFE || aligned) {
      const float4 v = ldg4(rowp + (SAFE ? min(xe, W - 4) : xe));
      b.e[0] = v.x; b.e[1] = v.y; b.e[2] = v.z; b.e[3] = v.w;
    } else {
#pragma unroll
      for (int t = 0; t < 4; ++t) b.e[t] = (sl < NE && xe + t < W) ? __ldg(rowp + xe + t) : 0.f;
    }
  }
}

// cp.async (LDGSTS) row ring: each lane copies its own quads global -> shared and later reads back
// only what it wrote itself, so deep prefetch costs no registers, no register copies and no
// cross-lane synchronisation (cp.async.wait_group per thread is enough).
__device__ __forceinline__ void cp_async16(unsigned saddr, const void *g) {
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(saddr), "l"(g) : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() {
  asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory");
}

// NST stages x (U+1) quads (U chunk quads + the halo quad) x 32 lanes x 16 B per warp
template <int K, int U, int SEG, int NST>
struct RowRing {
  static constexpr unsigned kStageBytes = (U + 1) * kWarp * 16;
  static constexpr unsigned kBytes = NST * kStageBytes;
  unsigned base;  // shared-window address of this warp's ring
  int lane, sl;

  // issue the copies of one row segment into `stage` (aligned rows; `clamp` on ragged edges)
  __device__ __forceinline__ void issue(int stage, const float *__restrict__ rowp, int x0, int W, bool clamp) const {
    constexpr int NE = KCfg<K>::NE;
    const unsigned sb = base + stage * kStageBytes + lane * 16;
#pragma unroll
    for (int u = 0; u < U; ++u) {
      int x = x0 + 4 * SEG * u + 4 * sl;
      if (clamp) x = min(x, W - 4);
      cp_async16(sb + u * kWarp * 16, rowp + x);
    }
    if constexpr (NE > 0) {
      int xe = x0 + 4 * SEG * U + 4 * (sl % NE);
      if (clamp) xe = min(xe, W - 4);
      cp_async16(sb + U * kWarp * 16, rowp + xe);
    }
    cp_async_commit();
  }
  __device__ __forceinline__ void read(int stage, RowBuf<K, U> &b) const {
    const unsigned sb = base + stage * kStageBytes + lane * 16;
#pragma unroll
    for (int u = 0; u < U; ++u) lds4_at(sb + u * kWarp * 16, b.a[u][0], b.a[u][1], b.a[u][2], b.a[u][3]);
    if constexpr (KCfg<K>::NE > 0) {
      lds4_at(sb + U * kWarp * 16, b.e[0], b.e[1], b.e[2], b.e[3]);
    } else {
#pragma unroll
      for (int t = 0; t < 4; ++t) b.e[t] = 0.f;
    }
  }
};

template <int K, int U, bool SAFE>
__device__ __forceinline__ void load_row(RowBuf<K, U> &b, const float *__restrict__ rowp, int x0, int W, int lane,
                                         bool aligned) {
  load_row_g<K, U, kWarp, SAFE>(b, rowp, x0, W, lane, aligned);
}

// ------------------------------------------------------------------------------------------------
// a2: column reuse -- assemble every chunk's window w[u][0..WN) = in[x0+4*SEG*u+4*sl .. +WN)
// ------------------------------------------------------------------------------------------------
// Halo element m (m = 4..K+2) of segment lane sl lives in register m%4 of segment lane sl + m/4.
// The SUPPLYING lane picks, with a static register index, its own register or -- if it is one of the
// first m/4 lanes, whose receivers wrap past the segment's last lane -- the next chunk's (or the halo
// quad's) register; one SEL + one SHFL.IDX (source lane inside the segment) per (m, chunk).
template <int K, int U, int SEG>
__device__ __forceinline__ void build_windows_g(const RowBuf<K, U> &b, float (&w)[U][KCfg<K>::WN], int lane) {
  const int sl = lane & (SEG - 1);
  const int base = lane & ~(SEG - 1);
#pragma unroll
  for (int u = 0; u < U; ++u) {
#pragma unroll
    for (int t = 0; t < 4; ++t) w[u][t] = b.a[u][t];
  }
#pragma unroll
  for (int m = 4; m < KCfg<K>::WN; ++m) {
    const int d = m >> 2;  // source lane offset (static)
    const int r = m & 3;   // source register (static)
    const int src = base | ((sl + d) & (SEG - 1));
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const float nxt = (u + 1 < U) ? b.a[(u + 1 < U) ? u + 1 : 0][r] : b.e[r];
      const float sup = (sl < d) ? nxt : b.a[u][r];
      w[u][m] = __shfl_sync(kFull, sup, src);
    }
  }
}

template <int K, int U>
__device__ __forceinline__ void build_windows(const RowBuf<K, U> &b, float (&w)[U][KCfg<K>::WN], int lane) {
  build_windows_g<K, U, kWarp>(b, w, lane);
}

// ------------------------------------------------------------------------------------------------
// a4: filter supply. A filter row i is fetched into K registers right before the FMAs that use it:
//   FSRC_CONST -- the __constant__ slot of this K (slot K, rows padded to KP floats), staged by the
//                 host with a stream-ordered 2D device-to-device copy; a call waits (stream-ordered,
//                 on a CUDA event) for the previous kernel that read the slot, so calls on other
//                 streams never see each other's filter. The slot address is a compile-time constant
//                 and the control flow is warp-uniform (one warp per CTA), so the compiler reads the
//                 filter with LDCU.128 into uniform registers and feeds FFMA's UR operand: one
//                 16-byte fetch per warp, no per-lane return traffic through the LSU/MIO path.
//   FSRC_SMEM  -- staged per CTA in shared memory (rows padded to KP floats), broadcast LDS.128. Each
//                 LDS.128 still returns 512 B through the shared-memory crossbar (16 B x 32 lanes),
//                 which caps large-K FMA throughput (profiles/); used when a launch is captured into
//                 a CUDA graph (the constant-slot recycling needs stream-ordered events).
// ------------------------------------------------------------------------------------------------
constexpr int FSRC_SMEM = 0;
constexpr int FSRC_CONST = 1;

constexpr int kConstSlotFloats = 256;  // >= 15 rows x 16 (padded) floats
// One slot per translation unit: every K is compiled in its own unit (csrc/inst_kNN.cu) and so in its
// own module with its own constant bank; slot "K" of the design is this array in unit K.
__constant__ __align__(16) float c_filt[kConstSlotFloats];

template <int K, int FSRC>
struct FilterSrc {
  unsigned sbase;      // FSRC_SMEM: shared-window address of row 0
  const float *cbase;  // FSRC_CONST: c_filt of this unit (compile-time address, rows of KP floats)

  __device__ __forceinline__ void row(float (&fr)[KCfg<K>::KP], int i) const {
    constexpr int KP = KCfg<K>::KP;
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

// ------------------------------------------------------------------------------------------------
// a6: store 4 outputs per lane of a 128-wide output chunk starting at g (16B alignment unknown)
// ------------------------------------------------------------------------------------------------
template <int S>
__device__ __forceinline__ void store_chunk_shifted(float *g, const float (&o)[4], int lane) {
  // g is S floats past a 16-byte boundary. Lanes 0..30 store the aligned quad at g + 4 - S + 4l:
  // own o[4-S..3] followed by lane l+1's o[0..3-S]. Lane 0 stores the 4-S head elements and lane 31
  // the S tail elements with scalar stores.
  float nb[4];
#pragma unroll
  for (int t = 0; t < 4; ++t) nb[t] = (t < 4 - S) ? __shfl_down_sync(kFull, o[t], 1) : 0.f;
  float q[4];
#pragma unroll
  for (int k = 0; k < 4; ++k) q[k] = (k < S) ? o[(4 - S + k) & 3] : nb[(k - S) & 3];
  if (lane < kWarp - 1) stg4(g + (4 - S) + 4 * lane, q[0], q[1], q[2], q[3]);
  if (lane == 0) {
#pragma unroll
    for (int t = 0; t < 4 - S; ++t) __stcs(g + t, o[t]);
  }
  if (lane == kWarp - 1) {
#pragma unroll
    for (int t = 4 - S; t < 4; ++t) __stcs(g + 4 * (kWarp - 1) + t, o[t]);
  }
}

// (A branch-free form -- all four realignments computed and selected, predicated head/tail
// stores -- measured slower on B200: 8192^2 K=7 388 vs 428 Gpx/s.)
__device__ __forceinline__ void store_chunk(float *g, const float (&o)[4], int lane) {
  const int s = static_cast<int>((reinterpret_cast<uintptr_t>(g) >> 2) & 3);
  switch (s) {  // warp-uniform: the dynamic shift becomes one of four static variants
    case 0: stg4(g + 4 * lane, o[0], o[1], o[2], o[3]); break;
    case 1: store_chunk_shifted<1>(g, o, lane); break;
    case 2: store_chunk_shifted<2>(g, o, lane); break;
    default: store_chunk_shifted<3>(g, o, lane); break;
  }
}

template <int U, bool SAFE>
__device__ __forceinline__ void store_row(float *__restrict__ orow, int x0, int Wo, const float (&o)[U][4],
                                          int lane) {
#pragma unroll
  for (int u = 0; u < U; ++u) {
    const int xb = x0 + 128 * u;
    if (!SAFE) {
      store_chunk(orow + xb, o[u], lane);
    } else {
#pragma unroll
      for (int t = 0; t < 4; ++t) {
        const int x = xb + 4 * lane + t;
        if (x < Wo) __stcs(orow + x, o[u][t]);
      }
    }
  }
}

// ------------------------------------------------------------------------------------------------
// a3: row reuse (single channel). acc[q] holds output row r-K+1+q after input row r.
// ------------------------------------------------------------------------------------------------
// One input row (windows w) into the ring: acc[q] = acc[q+1] + w . filter[K-1-q]. The ring shift is
// folded into the first FMA of each chain (no MOVs); per output the terms arrive in filter-row,
// filter-column order, independent of where the band starts (band-independent bits). GUARD: only
// slots qmin <= q < qmax -- the first K-1 rows of a band feed fewer of its outputs (Alg. 2 case 1),
// and so do the last K-1 (case 3); the branches are warp-uniform.
template <int K, int U, int FSRC, bool GUARD>
__device__ __forceinline__ void row_step1(float (&acc)[K][U][4], const float (&w)[U][KCfg<K>::WN],
                                          const FilterSrc<K, FSRC> &fs, int qmin, int qmax) {
  if constexpr (U == 2) {
    // Paired FMA (sm_100 FFMA2, fma.rn.f32x2) across the two column chunks: one instruction runs the
    // FMA chains of column v of chunk 0 and of chunk 1. Each component is an ordinary round-to-nearest
    // fp32 FMA, so every output's sum is the same sequence of fmaf steps as the scalar chain -- the
    // same bits -- but the FMA work takes half the issue slots (an FFMA2 = 64 FMAs occupies the FMA pipe
    // for 2 cycles and leaves the other issue cycle to the shuffles, filter fetches, loads and stores;
    // tools/ubench/ffma2_rate.cu: 99.8% of the fp32 peak vs 90-98% for FFMA). Every window value
    // belongs to exactly one (chunk 0, chunk 1) pair, so forming the pairs costs no copies (pairs of
    // adjacent columns (w[m], w[m+1]) straddle register pairs and cost ~200 MOVs per row at K=15); the
    // broadcast filter value (f, f) is FFMA2's scalar uniform-register operand.
#pragma unroll
    for (int q = 0; q < K; ++q) {
      if (!GUARD || (q >= qmin && q < qmax)) {
        float fr[KCfg<K>::KP];
        fs.row(fr, K - 1 - q);
#pragma unroll
        for (int v = 0; v < 4; ++v) {
          float2 s = (q + 1 < K) ? make_float2(acc[(q + 1 < K) ? q + 1 : 0][0][v], acc[(q + 1 < K) ? q + 1 : 0][1][v])
                                 : make_float2(0.f, 0.f);
#pragma unroll
          for (int j = 0; j < K; ++j)
            s = __ffma2_rn(make_float2(w[0][v + j], w[1][v + j]), make_float2(fr[j], fr[j]), s);
          acc[q][0][v] = s.x;
          acc[q][1][v] = s.y;
        }
      }
    }
  } else {
#pragma unroll
    for (int q = 0; q < K; ++q) {
      if (!GUARD || (q >= qmin && q < qmax)) {
        float fr[KCfg<K>::KP];
        fs.row(fr, K - 1 - q);
#pragma unroll
        for (int u = 0; u < U; ++u) {
#pragma unroll
          for (int v = 0; v < 4; ++v) {
            float s = (q + 1 < K) ? acc[(q + 1 < K) ? q + 1 : 0][u][v] : 0.f;
#pragma unroll
            for (int j = 0; j < K; ++j) s = fmaf(w[u][v + j], fr[j], s);
            acc[q][u][v] = s;
          }
        }
      }
    }
  }
}

// ------------------------------------------------------------------------------------------------
// Single-channel kernel
// ------------------------------------------------------------------------------------------------
struct SingleArgs {
  const float *in;
  const float *in2;  // rows >= H1 come from in2 (the halo of a row band, possibly a peer GPU's memory)
  int H1;            // rows [0, H1) at in, rows [H1, H) at in2 (H1 == H: one segment)
  int P;             // input row pitch in floats (>= W; == W for the C-ABI calls, padded buffers: % 4 == 0)
  int Wc;            // row-fetch bound: W, or P for a padded buffer (clamped quads stay in the pitch)
  int Po;            // output row pitch in floats (>= Wo; == Wo for the C-ABI calls)
  const float *filt;
  float *out;
  int H, W, Ho, Wo;
  int n_img;          // images of a batch (conv2d_single_batch); image i at in + i*img_in, out + i*img_out
  long long img_in;   // floats between consecutive input images (H * P)
  long long img_out;  // floats between consecutive output images (Ho * Po)
  int n_bands;        // output-row bands per image: band b = rows [b*Ho/n_bands, (b+1)*Ho/n_bands)
  int n_cb;           // column blocks of 128*U outputs
  int n_tiles;        // n_img * n_bands * n_cb
  int aligned;        // in is 16B aligned and W % 4 == 0
};

// Output rows of band b of n (balanced: heights differ by at most one row, so a wave of n_bands
// bands per column block is exactly n_bands tiles and no SM gets a short tile).
__device__ __forceinline__ int band_start(int b, int n, int Ho) {
  return static_cast<int>(static_cast<long long>(b) * Ho / n);
}

// HALO: rows >= H1 come from in2 (conv2d_single_halo); a separate instantiation, so the one-segment
// kernels keep their row addressing (the per-row select measured -2% at K = 11..15).
template <bool HALO>
__device__ __forceinline__ const float *in_row(const SingleArgs &a, const float *__restrict__ inb, int r) {
  if constexpr (HALO)
    return r < a.H1 ? inb + static_cast<size_t>(r) * a.P : a.in2 + static_cast<size_t>(r - a.H1) * a.P;
  else
    return inb + static_cast<size_t>(r) * a.P;
}

// One warp tile: 128*U columns x output rows [ob, oe). Input rows [ob, oe+K-1) stream through once,
// following Algorithm 2's three cases: the first K-1 rows feed only the slots of outputs
// >= ob (case 1, no stores), the steady state feeds all K slots and completes one output row per
// input row (case 2), the last K-1 rows feed only outputs < oe (case 3, fixed per DESIGN.md R8).
// GUARDS selects how cases 1 and 3 are run:
//   0 -- one loop, every row runs the full K-slot body (the extra FMAs of cases 1/3 land in slots that
//        are never stored): a single hot loop, no per-slot branches (best I-cache / scheduling);
//   1 -- case 1 in its own loop with per-slot warp-uniform branches, cases 2+3 unguarded;
//   2 -- cases 1 and 3 both guarded (no wasted FMA, but the per-slot branches split the FMA stream
//        into basic blocks the scheduler cannot overlap).
// Row r+1 (r+2 when PF == 2) is in flight from memory while row r is computed; the next-row index
// is clamped, so the loop body has no branch besides the store.
// EDGE 0: interior tile (vector loads / stores); 1: aligned rows, ragged right edge (clamped vector
// loads, masked scalar stores); 2: misaligned rows (guarded scalar loads, masked stores).
// PF 1/2: rows r+1 (r+2) in flight in registers; PF >= 3 (power of two, EDGE < 2): a PF-stage cp.async
// ring in shared memory with PF-1 rows in flight (latency-bound short bands and HBM-bound small K).
template <int K, int U, int FSRC, int PF, int GUARDS, int EDGE, bool HALO>
__device__ __forceinline__ void single_tile(const SingleArgs &a, const float *__restrict__ inb,
                                            float *__restrict__ outb, const FilterSrc<K, FSRC> &fs, int x0, int ob,
                                            int oe, int lane, unsigned ring_base) {
  constexpr bool SAFE = (EDGE != 0);
  constexpr int NST = (PF >= 3 && EDGE != 2) ? PF : 1;
  constexpr int RPF = (PF == 2 || (PF >= 3 && EDGE == 2)) ? ((PF == 2) ? 2 : 1) : 1;
  static_assert(NST == 1 || (NST & (NST - 1)) == 0, "ring depth must be a power of two");
  const int rend = oe + K - 1;  // input rows [ob, rend)
  const int rlast = rend - 1;
  float acc[K][U][4];
#pragma unroll
  for (int q = 0; q < K; ++q)
#pragma unroll
    for (int u = 0; u < U; ++u)
#pragma unroll
      for (int v = 0; v < 4; ++v) acc[q][u][v] = 0.f;
  RowRing<K, U, kWarp, (NST > 1 ? NST : 2)> ring;
  ring.base = ring_base;
  ring.lane = lane;
  ring.sl = lane;
  constexpr bool clamp = (EDGE == 1);
  RowBuf<K, U> n1, n2;  // register path: rows r+1 (and r+2 when RPF == 2) in flight
  if constexpr (NST > 1) {
#pragma unroll
    for (int st = 0; st < NST - 1; ++st) ring.issue(st, in_row<HALO>(a, inb, min(ob + st, rlast)), x0, a.Wc, clamp);
  } else {
    load_row<K, U, SAFE>(n1, in_row<HALO>(a, inb, ob), x0, a.Wc, lane, a.aligned);
    if (RPF == 2) load_row<K, U, SAFE>(n2, in_row<HALO>(a, inb, min(ob + 1, rlast)), x0, a.Wc, lane, a.aligned);
  }
  // returns row r and issues the fetch of row r+depth (index clamped)
  auto next_row = [&](int r) {
    RowBuf<K, U> cur;
    if constexpr (NST > 1) {
      cp_async_wait<NST - 2>();
      const int k = r - ob;
      ring.read(k & (NST - 1), cur);
      ring.issue((k + NST - 1) & (NST - 1), in_row<HALO>(a, inb, min(r + NST - 1, rlast)), x0, a.Wc, clamp);
    } else if constexpr (RPF == 2) {
      cur = n1;
      n1 = n2;
      load_row<K, U, SAFE>(n2, in_row<HALO>(a, inb, min(r + 2, rlast)), x0, a.Wc, lane, a.aligned);
    } else {
      cur = n1;
      load_row<K, U, SAFE>(n1, in_row<HALO>(a, inb, min(r + 1, rlast)), x0, a.Wc, lane, a.aligned);
    }
    return cur;
  };
  int r = ob;
  if constexpr (GUARDS == 0) {
    for (; r < rend; ++r) {
      const RowBuf<K, U> cur = next_row(r);
      float w[U][KCfg<K>::WN];
      build_windows<K, U>(cur, w, lane);
      row_step1<K, U, FSRC, false>(acc, w, fs, 0, K);
      if (r >= ob + K - 1) store_row<U, SAFE>(outb + static_cast<size_t>(r - K + 1) * a.Po, x0, a.Wo, acc[0], lane);
    }
    return;
  }
  for (; r < min(ob + K - 1, oe); ++r) {  // case 1: slots of outputs >= ob only
    const RowBuf<K, U> cur = next_row(r);
    float w[U][KCfg<K>::WN];
    build_windows<K, U>(cur, w, lane);
    row_step1<K, U, FSRC, true>(acc, w, fs, K - 1 - (r - ob), K);
  }
  const int steady_end = (GUARDS == 2) ? oe : rend;
  for (; r < steady_end; ++r) {  // case 2 (+3 when GUARDS == 1): all K slots
    const RowBuf<K, U> cur = next_row(r);
    float w[U][KCfg<K>::WN];
    build_windows<K, U>(cur, w, lane);
    row_step1<K, U, FSRC, false>(acc, w, fs, 0, K);
    if (GUARDS == 2 || r >= ob + K - 1) store_row<U, SAFE>(outb + static_cast<size_t>(r - K + 1) * a.Po, x0, a.Wo, acc[0], lane);
  }
  for (; r < rend; ++r) {  // case 3 (GUARDS == 2): slots of outputs < oe only (>= ob for short bands)
    const RowBuf<K, U> cur = next_row(r);
    float w[U][KCfg<K>::WN];
    build_windows<K, U>(cur, w, lane);
    row_step1<K, U, FSRC, true>(acc, w, fs, max(0, K - 1 - (r - ob)), oe + K - 1 - r);
    if (r >= ob + K - 1) store_row<U, SAFE>(outb + static_cast<size_t>(r - K + 1) * a.Po, x0, a.Wo, acc[0], lane);
  }
}

// CTAW: warps per CTA. With CTAW == 1 every branch depends only on blockIdx and kernel parameters,
// so the compiler can prove warp-uniform control flow and keep the constant-bank filter in uniform
// registers (LDCU + FFMA with UR operands) instead of per-lane loads.
// MINB > 1: resident CTAs per SM the register allocation must allow (ptxas otherwise picks its own cap).
template <int K, int U, int FSRC, int CTAW, int PF = 1, int GUARDS = 0, bool HALO = false, int MINB = 1>
__global__ void __launch_bounds__(CTAW *kWarp, MINB) k_conv2d_single(const SingleArgs a) {
  constexpr int KP = KCfg<K>::KP;
  __shared__ __align__(16) float sf[(FSRC == FSRC_SMEM) ? K * KP : 4];
  extern __shared__ __align__(16) float ring_smem[];  // PF >= 3: CTAW rings of RowRing::kBytes
  FilterSrc<K, FSRC> fs;
  if constexpr (FSRC == FSRC_CONST) {
    fs.cbase = c_filt;
  } else {
    for (int t = threadIdx.x; t < K * KP; t += blockDim.x) {
      const int i = t / KP, j = t % KP;
      sf[t] = (j < K) ? a.filt[i * K + j] : 0.f;
    }
    __syncthreads();
    fs.sbase = static_cast<unsigned>(__cvta_generic_to_shared(sf));
  }
  const int lane = threadIdx.x & (kWarp - 1);
  const int warp = (CTAW == 1) ? 0 : static_cast<int>(threadIdx.x >> 5);
  const int tile = static_cast<int>(blockIdx.x) * CTAW + warp;
  if (tile >= a.n_tiles) return;
  const unsigned ring_base = static_cast<unsigned>(__cvta_generic_to_shared(ring_smem)) +
                             warp * RowRing<K, U, kWarp, (PF >= 3 ? PF : 2)>::kBytes;
  const int cb = tile % a.n_cb;
  const int t2 = tile / a.n_cb;
  const int band = t2 % a.n_bands;
  const int img = t2 / a.n_bands;
  const float *__restrict__ inb = a.in + img * a.img_in;
  float *__restrict__ outb = a.out + img * a.img_out;
  const int x0 = cb * 128 * U;
  const int ob = band_start(band, a.n_bands, a.Ho);
  const int oe = band_start(band + 1, a.n_bands, a.Ho);
  // fast tiles: 16B-aligned rows, every column of the tile and its extra halo quad in range
  const bool inside = x0 + 128 * U + 4 * KCfg<K>::NE <= a.W;  // warp-uniform
  if (a.aligned && inside)
    single_tile<K, U, FSRC, PF, GUARDS, 0, HALO>(a, inb, outb, fs, x0, ob, oe, lane, ring_base);
  else if (a.aligned)
    single_tile<K, U, FSRC, PF, GUARDS, 1, HALO>(a, inb, outb, fs, x0, ob, oe, lane, ring_base);
  else
    single_tile<K, U, FSRC, PF, GUARDS, 2, HALO>(a, inb, outb, fs, x0, ob, oe, lane, ring_base);
}

// ------------------------------------------------------------------------------------------------
// Multi-channel kernel: FB filters per warp, C channels streamed per input row
// ------------------------------------------------------------------------------------------------
struct MultiArgs {
  const float *in;
  const float *filt;
  float *out;
  int N, C, H, W, F, Ho, Wo;
  int band_h, n_cb, n_bands, n_fb;
  long long n_tiles;
  int aligned;
};

// sfc: staged filters of channel c, layout [K][FB][KP] (filter row i of filter fb at (i*FB+fb)*KP)
template <int K, int FB, bool SHIFT>
__device__ __forceinline__ void row_reuse_multi(float (&acc)[K][FB][4], const float (&w)[KCfg<K>::WN],
                                                const float *__restrict__ sfc, int qmin) {
  constexpr int KP = KCfg<K>::KP;
#pragma unroll
  for (int q = 0; q < K; ++q) {
    if (q >= qmin) {
      const int i = K - 1 - q;
#pragma unroll
      for (int fb = 0; fb < FB; ++fb) {
        float fr[KP];
#pragma unroll
        for (int c4 = 0; c4 < KP / 4; ++c4)
          lds4_volatile(sfc + (i * FB + fb) * KP + 4 * c4, fr[4 * c4], fr[4 * c4 + 1], fr[4 * c4 + 2],
                        fr[4 * c4 + 3]);
#pragma unroll
        for (int v = 0; v < 4; ++v) {
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

template <int K, int FB, bool SAFE>
__device__ __forceinline__ void multi_tile(const MultiArgs &a, const float *__restrict__ sf, int n, int f0,
                                           int x0, int ob, int oe, int lane) {
  constexpr int KP = KCfg<K>::KP;
  const int rend = oe + K - 1;
  const int C = a.C;
  const size_t plane = static_cast<size_t>(a.H) * a.W;
  const float *__restrict__ img = a.in + static_cast<size_t>(n) * C * plane;

  float acc[K][FB][4];
#pragma unroll
  for (int q = 0; q < K; ++q)
#pragma unroll
    for (int fb = 0; fb < FB; ++fb)
#pragma unroll
      for (int v = 0; v < 4; ++v) acc[q][fb][v] = 0.f;

  RowBuf<K, 1> nxt;
  load_row<K, 1, SAFE>(nxt, img + static_cast<size_t>(ob) * a.W, x0, a.W, lane, a.aligned);
  for (int r = ob; r < rend; ++r) {
    const int done = r - ob;
    const int qmin = (done < K - 1) ? (K - 1 - done) : 0;
    for (int c = 0; c < C; ++c) {
      RowBuf<K, 1> cur = nxt;
      // prefetch the next (row, channel) of the stream
      {
        int rn = r, cn = c + 1;
        if (cn == C) { cn = 0; ++rn; }
        if (rn < rend)
          load_row<K, 1, SAFE>(nxt, img + cn * plane + static_cast<size_t>(rn) * a.W, x0, a.W, lane, a.aligned);
      }
      float w[1][KCfg<K>::WN];
      build_windows<K, 1>(cur, w, lane);
      const float *sfc = sf + static_cast<size_t>(c) * K * FB * KP;
      if (c == 0)
        row_reuse_multi<K, FB, true>(acc, w[0], sfc, qmin);
      else
        row_reuse_multi<K, FB, false>(acc, w[0], sfc, qmin);
    }
    if (done >= K - 1) {
      const int o = r - K + 1;
#pragma unroll
      for (int fb = 0; fb < FB; ++fb) {
        if (f0 + fb < a.F) {
          float *orow = a.out + ((static_cast<size_t>(n) * a.F + f0 + fb) * a.Ho + o) * a.Wo;
          float ov[1][4];
#pragma unroll
          for (int v = 0; v < 4; ++v) ov[0][v] = acc[0][fb][v];
          store_row<1, SAFE>(orow, x0, a.Wo, ov, lane);
        }
      }
    }
  }
}

template <int K, int FB>
// (the explicit 2 CTAs/SM keeps ptxas from capping the registers at 96 and spilling: tests/test_sass.py)
__global__ void __launch_bounds__(kCtaWarps *kWarp, 2) k_conv2d_multi(const MultiArgs a) {
  constexpr int KP = KCfg<K>::KP;
  extern __shared__ __align__(16) float smem[];
  // CTA = 4 warps on the same (n, F-block): stage that block's filters, layout [C][K][FB][KP]
  const long long cta_tile0 = static_cast<long long>(blockIdx.x) * kCtaWarps;
  const long long per_fb = static_cast<long long>(a.n_cb) * a.n_bands;  // tiles per (n, F-block)
  const int fblk = static_cast<int>((cta_tile0 / per_fb) % a.n_fb);
  // host guarantees per_fb % kCtaWarps == 0, so all warps of the CTA share (n, fblk)
  const int f0 = fblk * FB;
  const int C = a.C;
  const int total = C * K * FB * KP;
  for (int t = threadIdx.x; t < total; t += blockDim.x) {
    const int j = t % KP;
    const int fb = (t / KP) % FB;
    const int i = (t / (KP * FB)) % K;
    const int c = t / (KP * FB * K);
    const int f = f0 + fb;
    smem[t] = (j < K && f < a.F) ? a.filt[((static_cast<size_t>(f) * C + c) * K + i) * K + j] : 0.f;
  }
  __syncthreads();

  const int lane = threadIdx.x & (kWarp - 1);
  const long long tile = cta_tile0 + (threadIdx.x >> 5);
  if (tile >= a.n_tiles) return;
  const int cb = static_cast<int>(tile % a.n_cb);
  const int band = static_cast<int>((tile / a.n_cb) % a.n_bands);
  const int n = static_cast<int>(tile / (per_fb * a.n_fb));
  const int x0 = cb * 128;
  const int ob = band * a.band_h;
  const int oe = min(ob + a.band_h, a.Ho);
  if (ob >= a.Ho) return;
  const bool fast = a.aligned && (x0 + 128 + 4 * KCfg<K>::NE <= a.W);
  if (fast)
    multi_tile<K, FB, false>(a, smem, n, f0, x0, ob, oe, lane);
  else
    multi_tile<K, FB, true>(a, smem, n, f0, x0, ob, oe, lane);
}

}  // namespace c2d

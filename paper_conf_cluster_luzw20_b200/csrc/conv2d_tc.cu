// conv2d_tc.cu -- tensor-core variant of the multi-channel convolution: the large-C
// case is a dense contraction, D[p][f] = sum_k A[p][k] * B[k][f] with p output pixels, f filters and
// k = (c, i, j), A[p][k] = in[n][c][y+i][x+j] (implicit im2col), B[k][f] = w[f][c][i][j].
// It runs on the 5th-generation tensor cores (tcgen05.mma kind::tf32, accumulator in TMEM) with the
// 3xTF32 split a = a_hi + a_lo (a_hi = tf32(a) rounded to nearest, a_lo = a - a_hi exact in fp32):
//     D = A_hi B_hi + A_hi B_lo + A_lo B_hi      (the dropped A_lo B_lo term is ~2^-22 |a||b|)
// which keeps each product within ~2^-21 relative, far inside the 1e-5 * sum|x||w| acceptance
// (DESIGN.md "Tensor-core variant"). A separate, measured variant, as BASELINE.json north_star asks.
//
// Design (v2):
//   * Pixels are indexed with the INPUT row pitch, p = y*W + x (x < W, not Wo): for a fixed
//     k = (c, i, j) the A column of 128 consecutive pixels is then 128 consecutive input floats at
//     plane offset p0 + i*W + j, so every gather is one coalesced 128-byte warp load. The W-Wo pixels
//     per row with x >= Wo are computed from clamped addresses and never stored.
//   * A (im2col) goes straight from registers to TMEM (tcgen05.st), never through shared memory:
//     a gather thread owns one pixel row = one TMEM lane, splits its 16 k-values of a K block into
//     hi/lo and stores them into the 32 + 32 TMEM columns of an A stage; the MMA reads A from
//     TMEM ("TS" form) and only B from shared memory. This removes the A shared-memory round trip and
//     the A re-reads that made the first version shared-memory bound.
//   * B (filters) is split once per call by a small kernel into hi/lo tiles laid out exactly as the
//     canonical K-major no-swizzle UMMA shared-memory image of each (filter block, K block); a
//     producer thread streams them with 1-D bulk copies (cp.async.bulk, mbarrier complete_tx) into a
//     deeper ring than A, so B latency is off the critical path.
//   * Warp roles (320 threads): warps 0-7 gather A and run the epilogue (warps w and w+4 share TMEM
//     lane quarter w%4 and take one half of each K block's 32 k), warp 8 allocates TMEM and one lane
//     issues the MMAs (12 per K block: 4 k-steps x 3 split products) and commits them to the stage
//     "empty" barriers, warp 9 lane 0 produces B. Global loads of K blocks kb+1 and kb+2 are in
//     flight in registers while block kb is split and stored.
//   * Epilogue: tcgen05.ld (each warp its 32 TMEM lanes) -> NFHoWo stores, coalesced along pixels.
#include <atomic>
#include <cstdint>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"
#include "common.h"

namespace c2d_tc {

constexpr int kM = 128;        // pixels per tile (UMMA M, TMEM lanes)
constexpr int kKB = 32;        // k values per K block (4 UMMA K=8 steps)
constexpr int kGather = 256;   // gather / epilogue threads (warps 0-7: two per TMEM lane quarter)
constexpr int kMmaWarp = 8;    // TMEM allocation + MMA issue
constexpr int kProdWarp = 9;   // B producer
constexpr int kThreads = 320;
constexpr int kKH = kKB / 2;   // k values per gather thread and K block

__device__ __forceinline__ uint32_t smem_u32(const void *p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

__host__ __device__ constexpr int tile_elem(int rows, int r, int k) {
  // element (row r, k) of a [rows x 32] K-major no-swizzle tile: core matrix (k/4, r/8) of 8 rows x 16 B
  return ((k >> 2) * (rows >> 3) + (r >> 3)) * 32 + (r & 7) * 4 + (k & 3);
}

__device__ __forceinline__ float tf32_hi(float a) {
  uint32_t r;
  asm("cvt.rna.tf32.f32 %0, %1;" : "=r"(r) : "f"(a));
  return __uint_as_float(r);
}

// round-to-nearest (ties away) to the tf32 grid on the bit pattern: 2 integer ops instead of the
// Inf/NaN-guarded cvt.rna sequence. Equal to cvt.rna.tf32 for every finite |a| < 0x1.ffep127 and for
// +-Inf / NaN (the carry never leaves the exponent field there).
__device__ __forceinline__ float tf32_hi_fast(float a) {
  return __uint_as_float((__float_as_uint(a) + 0x1000u) & 0xffffe000u);
}

// canonical K-major, SWIZZLE_NONE UMMA shared-memory descriptor (cute::UMMA::SmemDescriptor layout):
// start>>4 [0,14), LBO>>4 [16,30) = stride between the two 16-byte K chunks of an 8-row core
// matrix group, SBO>>4 [32,46) = stride between 8-row groups, version 1 [46,48), layout 0 [61,64)
__device__ __forceinline__ uint64_t umma_desc(uint32_t saddr, uint32_t lbo, uint32_t sbo) {
  uint64_t d = 0;
  d |= static_cast<uint64_t>((saddr >> 4) & 0x3FFF);
  d |= static_cast<uint64_t>((lbo >> 4) & 0x3FFF) << 16;
  d |= static_cast<uint64_t>((sbo >> 4) & 0x3FFF) << 32;
  d |= static_cast<uint64_t>(1) << 46;
  return d;
}

// instruction descriptor, kind::tf32: D f32, A/B tf32, both K-major, N>>3 at [17,23), M>>4 at [24,29)
__host__ __device__ constexpr uint32_t idesc_tf32(int M, int N) {
  return (1u << 4) | (2u << 7) | (2u << 10) | (static_cast<uint32_t>(N >> 3) << 17) |
         (static_cast<uint32_t>(M >> 4) << 24);
}

// D (TMEM) (+)= A (TMEM) x B (shared memory descriptor)
__device__ __forceinline__ void mma_tf32_ts(uint32_t tmem_d, uint32_t tmem_a, uint64_t bdesc, uint32_t idesc,
                                            uint32_t accumulate) {
  asm volatile(
      "{\n\t.reg .pred p;\n\t"
      "setp.ne.b32 p, %4, 0;\n\t"
      "tcgen05.mma.cta_group::1.kind::tf32 [%0], [%1], %2, %3, p;\n\t}\n" ::"r"(tmem_d),
      "r"(tmem_a), "l"(bdesc), "r"(idesc), "r"(accumulate));
}

__device__ __forceinline__ void mma_commit(uint32_t mbar) {
  asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(mbar)
               : "memory");
}

__device__ __forceinline__ void mbar_init(uint32_t mbar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(mbar), "r"(count) : "memory");
}

__device__ __forceinline__ void mbar_arrive(uint32_t mbar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(mbar) : "memory");
}

__device__ __forceinline__ void mbar_arrive_tx(uint32_t mbar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(mbar), "r"(bytes) : "memory");
}

__device__ __forceinline__ void mbar_wait(uint32_t mbar, uint32_t parity) {
  asm volatile(
      "{\n\t.reg .pred done;\n\t"
      "WAIT_%=:\n\t"
      "mbarrier.try_wait.parity.shared::cta.b64 done, [%0], %1;\n\t"
      "@!done bra WAIT_%=;\n\t}\n" ::"r"(mbar),
      "r"(parity)
      : "memory");
}

__device__ __forceinline__ void bulk_g2s(uint32_t dst, const void *src, uint32_t bytes, uint32_t mbar) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(dst),
               "l"(src), "r"(bytes), "r"(mbar)
               : "memory");
}

__device__ __forceinline__ void tc_fence_before() { asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory"); }
__device__ __forceinline__ void tc_fence_after() { asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory"); }

__device__ __forceinline__ void tmem_st32(uint32_t taddr, const uint32_t (&r)[32]) {
  asm volatile(
      "tcgen05.st.sync.aligned.32x32b.x32.b32 [%0], {%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,%16,"
      "%17,%18,%19,%20,%21,%22,%23,%24,%25,%26,%27,%28,%29,%30,%31,%32};" ::"r"(taddr),
      "r"(r[0]), "r"(r[1]), "r"(r[2]), "r"(r[3]), "r"(r[4]), "r"(r[5]), "r"(r[6]), "r"(r[7]), "r"(r[8]), "r"(r[9]),
      "r"(r[10]), "r"(r[11]), "r"(r[12]), "r"(r[13]), "r"(r[14]), "r"(r[15]), "r"(r[16]), "r"(r[17]), "r"(r[18]),
      "r"(r[19]), "r"(r[20]), "r"(r[21]), "r"(r[22]), "r"(r[23]), "r"(r[24]), "r"(r[25]), "r"(r[26]), "r"(r[27]),
      "r"(r[28]), "r"(r[29]), "r"(r[30]), "r"(r[31])
      : "memory");
}

__device__ __forceinline__ void tmem_st16(uint32_t taddr, const uint32_t (&r)[16]) {
  asm volatile(
      "tcgen05.st.sync.aligned.32x32b.x16.b32 [%0], {%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,%16};" ::"r"(
          taddr),
      "r"(r[0]), "r"(r[1]), "r"(r[2]), "r"(r[3]), "r"(r[4]), "r"(r[5]), "r"(r[6]), "r"(r[7]), "r"(r[8]), "r"(r[9]),
      "r"(r[10]), "r"(r[11]), "r"(r[12]), "r"(r[13]), "r"(r[14]), "r"(r[15])
      : "memory");
}

__device__ __forceinline__ void tmem_st8(uint32_t taddr, const uint32_t (&r)[8]) {
  asm volatile("tcgen05.st.sync.aligned.32x32b.x8.b32 [%0], {%1,%2,%3,%4,%5,%6,%7,%8};" ::"r"(taddr), "r"(r[0]),
               "r"(r[1]), "r"(r[2]), "r"(r[3]), "r"(r[4]), "r"(r[5]), "r"(r[6]), "r"(r[7])
               : "memory");
}

template <int NV>
__device__ __forceinline__ void tmem_stv(uint32_t taddr, const uint32_t (&r)[NV]) {
  if constexpr (NV == 16) {
    tmem_st16(taddr, r);
  } else {
    static_assert(NV == 8, "8 or 16 columns");
    tmem_st8(taddr, r);
  }
}

__device__ __forceinline__ void tmem_ld16(uint32_t taddr, float (&v)[16]) {
  uint32_t r[16];
  asm volatile(
      "tcgen05.ld.sync.aligned.32x32b.x16.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15}, [%16];"
      : "=r"(r[0]), "=r"(r[1]), "=r"(r[2]), "=r"(r[3]), "=r"(r[4]), "=r"(r[5]), "=r"(r[6]), "=r"(r[7]),
        "=r"(r[8]), "=r"(r[9]), "=r"(r[10]), "=r"(r[11]), "=r"(r[12]), "=r"(r[13]), "=r"(r[14]), "=r"(r[15])
      : "r"(taddr));
  asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
#pragma unroll
  for (int i = 0; i < 16; ++i) v[i] = __uint_as_float(r[i]);
}

// ------------------------------------------------------------------------------------------------
// filter split: Bs[fb][kb] = { hi tile [FN x 32], lo tile [FN x 32] } in the UMMA shared-memory image
// ------------------------------------------------------------------------------------------------
__global__ void k_tc_split_filters(const float *__restrict__ filt, int F, int Kg, int FN, int n_kb, int n_fb,
                                   float *__restrict__ bs) {
  const long long total = static_cast<long long>(n_fb) * n_kb * FN * kKB;
  for (long long e = static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x; e < total;
       e += static_cast<long long>(gridDim.x) * blockDim.x) {
    const int k = static_cast<int>(e % kKB);
    const int f = static_cast<int>((e / kKB) % FN);
    const int kb = static_cast<int>((e / (kKB * FN)) % n_kb);
    const int fb = static_cast<int>(e / (static_cast<long long>(kKB) * FN * n_kb));
    const int fg = fb * FN + f, kg = kb * kKB + k;
    const float v = (fg < F && kg < Kg) ? filt[static_cast<size_t>(fg) * Kg + kg] : 0.f;
    const float hi = tf32_hi(v);
    float *tile = bs + (static_cast<size_t>(fb) * n_kb + kb) * 2 * FN * kKB;
    tile[tile_elem(FN, f, k)] = hi;
    tile[FN * kKB + tile_elem(FN, f, k)] = v - hi;
  }
}

// ------------------------------------------------------------------------------------------------
// main kernel
// ------------------------------------------------------------------------------------------------
struct TcArgs {
  const float *in;
  const float *bs;  // split filters (k_tc_split_filters)
  float *out;
  int N, C, H, W, F, K, Ho, Wo;
  int Kg;             // C * K * K
  int n_kb;           // K blocks of 32
  int tiles_per_img;  // ceil(Ho * W / 128)
};

// NBS: B ring depth selector (0 = default; otherwise the stage count, for tuning)
// NACC: 1 = one accumulator; 2 = A_hi B_hi into accumulator 0 and the two correction products into
// accumulator 1 (summed in the epilogue) -- two independent MMA dependency chains per CTA
template <int FN, int NBS = 0, int NACC = 1>
struct TcCfg {
  static constexpr int NSA = NACC == 1 ? ((FN <= 64) ? 3 : (FN <= 128 ? 2 : 4))
                                       : ((FN <= 32) ? 3 : (FN <= 64 ? 2 : 4));  // A stages (TMEM, 64 cols)
  static constexpr uint32_t kBStage = 2u * FN * kKB * 4u;            // B hi + lo tile bytes
  static constexpr int NSB = NBS ? NBS : ((FN <= 32) ? 8 : (FN <= 64 ? 6 : 3));  // B stages (smem)
  static constexpr int kAcc = NACC * FN;
  static constexpr int kCols = kAcc + NSA * 2 * kKB;                 // TMEM columns used
  static constexpr int kAlloc = kCols <= 32 ? 32 : kCols <= 64 ? 64 : kCols <= 128 ? 128 : kCols <= 256 ? 256 : 512;
};

template <int FN, int D, int NBS, int NACC>
__global__ void __launch_bounds__(kThreads, 2) k_conv2d_multi_tc4(const TcArgs a) {
  using Cfg = TcCfg<FN, NBS, NACC>;
  constexpr int NSA = Cfg::NSA, NSB = Cfg::NSB;
  extern __shared__ __align__(1024) uint8_t smem[];  // [NSB B stages] + int koff[n_kb * 32]
  __shared__ __align__(8) uint64_t full_a[NSA], empty_a[NSA], full_b[NSB], empty_b[NSB], acc_full;
  __shared__ uint32_t tmem_base_s;
  const int tid = threadIdx.x;
  const int warp = tid >> 5;
  const int lane = tid & 31;
  int *koff = reinterpret_cast<int *>(smem + NSB * Cfg::kBStage);

  if (warp == kMmaWarp) {  // TMEM: accumulator [0, FN) + NSA A stages of 64 columns
    asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(&tmem_base_s)),
                 "r"(Cfg::kAlloc));
    asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
  }
  if (tid == 0) {
    for (int s = 0; s < NSA; ++s) {
      mbar_init(smem_u32(&full_a[s]), kGather);
      mbar_init(smem_u32(&empty_a[s]), 1);
    }
    for (int s = 0; s < NSB; ++s) {
      mbar_init(smem_u32(&full_b[s]), 1);
      mbar_init(smem_u32(&empty_b[s]), 1);
    }
    mbar_init(smem_u32(&acc_full), 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  // im2col offsets of every k = (c, i, j) relative to the pixel's (c=0, y, x) input element; the
  // padding k >= Kg point at offset 0 (always in range; their B entries are zero)
  const int KK0 = a.K * a.K;
  const int plane = a.H * a.W;
  for (int k = tid; k < a.n_kb * kKB; k += kThreads) {
    int o = 0;
    if (k < a.Kg) {
      const int c = k / KK0, ij = k - c * KK0;
      const int i = ij / a.K, j = ij - i * a.K;
      o = c * plane + i * a.W + j;
    }
    koff[k] = o;
  }
  tc_fence_before();
  __syncthreads();
  tc_fence_after();
  const uint32_t tmem = tmem_base_s;
  const int n = blockIdx.x / a.tiles_per_img;
  const int t = blockIdx.x - n * a.tiles_per_img;
  const int fblk = blockIdx.y;
  const uint32_t sb_base = smem_u32(smem);

  if (warp < 8) {
    // ---------------- gather: pixel p = y*W + x of image n ----------------
    // warp w serves TMEM lane quarter w%4 (pixel rows 32(w%4)..+31) and k half w/4 of every K block
    const int quarter = warp & 3, khalf = warp >> 2;
    const int row = quarter * 32 + lane;
    const int pp = t * kM + row;
    const int y = pp / a.W, x = pp - y * a.W;
    const bool valid = (y < a.Ho) && (x < a.Wo);
    const int pe = valid ? pp : 0;  // garbage pixels read pixel 0's window (in range)
    const float *__restrict__ img = a.in + static_cast<size_t>(n) * a.C * plane + pe;
    const uint32_t t_lane = static_cast<uint32_t>(quarter * 32) << 16;

    auto load = [&](float (&v)[kKH], int kb) {
      const int4 *ko = reinterpret_cast<const int4 *>(koff + kb * kKB + khalf * kKH);
#pragma unroll
      for (int q = 0; q < kKH / 4; ++q) {
        const int4 o = ko[q];
        v[4 * q + 0] = __ldg(img + o.x);
        v[4 * q + 1] = __ldg(img + o.y);
        v[4 * q + 2] = __ldg(img + o.z);
        v[4 * q + 3] = __ldg(img + o.w);
      }
    };
    auto put = [&](float (&v)[kKH], int kb) {
      const int s = kb % NSA;
      if (kb >= NSA) {
        mbar_wait(smem_u32(&empty_a[s]), static_cast<uint32_t>((kb / NSA - 1) & 1));
        tc_fence_after();
      }
      if (kb == a.n_kb - 1) {  // padding k >= Kg: exact zeros (no Inf/NaN from the clamped reads)
#pragma unroll
        for (int q = 0; q < kKH; ++q)
          if (kb * kKB + khalf * kKH + q >= a.Kg) v[q] = 0.f;
      }
      uint32_t hi[kKH], lo[kKH];
#pragma unroll
      for (int q = 0; q < kKH; ++q) {
        const float h = tf32_hi_fast(v[q]);
        hi[q] = __float_as_uint(h);
        lo[q] = __float_as_uint(v[q] - h);
      }
      const uint32_t col = tmem + t_lane + Cfg::kAcc + s * 2 * kKB + khalf * kKH;
      tmem_st16(col, hi);
      tmem_st16(col + kKB, lo);
      asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
      tc_fence_before();
      mbar_arrive(smem_u32(&full_a[s]));
    };
    // ring of D register buffers: the loads of K blocks kb+1 .. kb+D-1 are in flight while block kb
    // is split and stored
    float v[D][kKH];
#pragma unroll
    for (int d = 0; d < D; ++d)
      if (d < a.n_kb) load(v[d], d);
    for (int kb0 = 0; kb0 < a.n_kb; kb0 += D) {
#pragma unroll
      for (int d = 0; d < D; ++d) {
        const int kb = kb0 + d;
        if (kb < a.n_kb) {
          put(v[d], kb);
          if (kb + D < a.n_kb) load(v[d], kb + D);
        }
      }
    }

    // ---------------- epilogue: TMEM accumulator -> out[n][f][y][x] ----------------
    mbar_wait(smem_u32(&acc_full), 0);
    tc_fence_after();
    const size_t PP = static_cast<size_t>(a.Ho) * a.Wo;
    float *__restrict__ obase = a.out + (static_cast<size_t>(n) * a.F) * PP + (valid ? (y * a.Wo + x) : 0);
    const int f0 = fblk * FN;
#pragma unroll 1
    for (int c0 = khalf * (FN / 2); c0 < (khalf + 1) * (FN / 2); c0 += 16) {
      float v[16];
      tmem_ld16(tmem + t_lane + c0, v);
      if constexpr (NACC == 2) {
        float c[16];
        tmem_ld16(tmem + t_lane + FN + c0, c);
#pragma unroll
        for (int q = 0; q < 16; ++q) v[q] += c[q];
      }
      if (valid) {
#pragma unroll
        for (int q = 0; q < 16; ++q) {
          const int f = f0 + c0 + q;
          if (f < a.F) __stcs(obase + static_cast<size_t>(f) * PP, v[q]);
        }
      }
    }
  } else if (warp == kMmaWarp) {
    // ---------------- MMA issuer ----------------
    if (lane == 0) {
      constexpr uint32_t idesc = idesc_tf32(kM, FN);
      constexpr uint32_t lbo = (FN / 8) * 128;
      for (int kb = 0; kb < a.n_kb; ++kb) {
        const int sa = kb % NSA, sb = kb % NSB;
        mbar_wait(smem_u32(&full_a[sa]), static_cast<uint32_t>((kb / NSA) & 1));
        mbar_wait(smem_u32(&full_b[sb]), static_cast<uint32_t>((kb / NSB) & 1));
        tc_fence_after();
        const uint32_t a_hi = tmem + Cfg::kAcc + sa * 2 * kKB, a_lo = a_hi + kKB;
        const uint32_t b_hi = sb_base + sb * Cfg::kBStage, b_lo = b_hi + Cfg::kBStage / 2;
        const uint32_t d1 = tmem + (NACC == 2 ? FN : 0);  // accumulator of the correction products
#pragma unroll
        for (int kk = 0; kk < kKB / 8; ++kk) {
          const uint32_t bo = static_cast<uint32_t>(2 * kk * (FN / 8) * 128);
          const uint64_t dbh = umma_desc(b_hi + bo, lbo, 128), dbl = umma_desc(b_lo + bo, lbo, 128);
          const uint32_t acc0 = (kb > 0 || kk > 0) ? 1u : 0u;
          mma_tf32_ts(tmem, a_hi + 8 * kk, dbh, idesc, acc0);
          mma_tf32_ts(d1, a_hi + 8 * kk, dbl, idesc, NACC == 2 ? acc0 : 1u);
          mma_tf32_ts(d1, a_lo + 8 * kk, dbh, idesc, 1u);
        }
        mma_commit(smem_u32(&empty_a[sa]));
        mma_commit(smem_u32(&empty_b[sb]));
      }
      mma_commit(smem_u32(&acc_full));
    }
  } else {
    // ---------------- B producer: bulk copies of the split filter tiles ----------------
    if (lane == 0) {
      const float *src = a.bs + static_cast<size_t>(fblk) * a.n_kb * (Cfg::kBStage / 4);
      for (int kb = 0; kb < a.n_kb; ++kb) {
        const int sb = kb % NSB;
        if (kb >= NSB) mbar_wait(smem_u32(&empty_b[sb]), static_cast<uint32_t>((kb / NSB - 1) & 1));
        mbar_arrive_tx(smem_u32(&full_b[sb]), Cfg::kBStage);
        bulk_g2s(sb_base + sb * Cfg::kBStage, src + static_cast<size_t>(kb) * (Cfg::kBStage / 4), Cfg::kBStage,
                 smem_u32(&full_b[sb]));
      }
    }
  }
  tc_fence_before();
  __syncthreads();
  if (warp == kMmaWarp) {
    tc_fence_after();
    asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(Cfg::kAlloc));
  }
}

// ------------------------------------------------------------------------------------------------
// persistent kernel: one CTA per SM walks the tiles (pixel tile x filter block) of the launch; two
// TMEM accumulators let the epilogue of tile j run on dedicated warps while the MMAs of tile j+1
// accumulate into the other buffer, and the A / B rings run continuously across tile boundaries
// ------------------------------------------------------------------------------------------------
// warps [0, GW): A gather (GW/4 per TMEM lane quarter, each a 32*4/GW-wide k slice of every K
// block); [GW, GW+4): epilogue; GW+4: TMEM allocation + MMA issue; GW+5: B producer
template <int GW>
struct TcPWarps {
  static constexpr int kGather = GW * 32;
  static constexpr int kEpi0 = GW;
  static constexpr int kMma = GW + 4;
  static constexpr int kProd = GW + 5;
  static constexpr int kThreads = (GW + 6) * 32;
  static constexpr int kKS = kKB * 4 / GW;  // k values per gather thread and K block
};

template <int FN>
struct TcPCfg {
  static constexpr int NSA = 4;                          // A stages (TMEM, 64 columns each)
  static constexpr uint32_t kBStage = 2u * FN * kKB * 4u;  // B hi + lo tile bytes
  static constexpr int NSB = (FN <= 64) ? 8 : 4;         // B stages (shared memory, 128 KB)
  static constexpr int kAcc = 2 * FN;                    // two accumulators
  static constexpr int kCols = kAcc + NSA * 2 * kKB;
  static_assert(kCols <= 512, "TMEM");
  static constexpr int kAlloc = kCols <= 256 ? 256 : 512;
};

struct TcTile {
  int n, t, fblk;
};

__device__ __forceinline__ TcTile tc_tile(const TcArgs &a, int n_fb, int tile) {
  TcTile r;
  const int pt = tile / n_fb;  // filter blocks innermost: consecutive tiles share their pixels
  r.fblk = tile - pt * n_fb;
  r.n = pt / a.tiles_per_img;
  r.t = pt - r.n * a.tiles_per_img;
  return r;
}

template <int FN, int D, int GW>
__global__ void __launch_bounds__(TcPWarps<GW>::kThreads, 1) k_conv2d_multi_tc5(const TcArgs a, int n_fb, int n_tiles) {
  using Cfg = TcPCfg<FN>;
  using Wp = TcPWarps<GW>;
  constexpr int KS = Wp::kKS;
  constexpr int NSA = Cfg::NSA, NSB = Cfg::NSB;
  extern __shared__ __align__(1024) uint8_t smem[];  // [NSB B stages] + int koff[n_kb * 32]
  __shared__ __align__(8) uint64_t full_a[NSA], empty_a[NSA], full_b[NSB], empty_b[NSB], acc_full[2],
      acc_empty[2];
  __shared__ uint32_t tmem_base_s;
  const int tid = threadIdx.x;
  const int warp = tid >> 5;
  const int lane = tid & 31;
  int *koff = reinterpret_cast<int *>(smem + NSB * Cfg::kBStage);

  if (warp == Wp::kMma) {
    asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(&tmem_base_s)),
                 "r"(Cfg::kAlloc));
    asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
  }
  if (tid == 0) {
    for (int s = 0; s < NSA; ++s) {
      mbar_init(smem_u32(&full_a[s]), Wp::kGather);
      mbar_init(smem_u32(&empty_a[s]), 1);
    }
    for (int s = 0; s < NSB; ++s) {
      mbar_init(smem_u32(&full_b[s]), 1);
      mbar_init(smem_u32(&empty_b[s]), 1);
    }
    for (int b = 0; b < 2; ++b) {
      mbar_init(smem_u32(&acc_full[b]), 1);
      mbar_init(smem_u32(&acc_empty[b]), 128);
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  const int KK0 = a.K * a.K;
  const int plane = a.H * a.W;
  for (int k = tid; k < a.n_kb * kKB; k += Wp::kThreads) {
    int o = 0;
    if (k < a.Kg) {
      const int c = k / KK0, ij = k - c * KK0;
      const int i = ij / a.K, j = ij - i * a.K;
      o = c * plane + i * a.W + j;
    }
    koff[k] = o;
  }
  tc_fence_before();
  __syncthreads();
  tc_fence_after();
  const uint32_t tmem = tmem_base_s;
  const uint32_t sb_base = smem_u32(smem);
  // this CTA's tiles: blockIdx.x, blockIdx.x + gridDim.x, ...; local block stream g = j * n_kb + kb
  const int my_tiles = (n_tiles - static_cast<int>(blockIdx.x) + static_cast<int>(gridDim.x) - 1) /
                       static_cast<int>(gridDim.x);
  const int n_blocks = my_tiles * a.n_kb;
  // small filter banks (one filter block, K blocks <= ring stages) are loaded once and stay resident
  const bool b_resident = (n_fb == 1) && (a.n_kb <= NSB);

  if (warp < GW) {
    // ---------------- gather (A producer) ----------------
    const int quarter = warp & 3, kpart = warp >> 2;
    const int row = quarter * 32 + lane;
    const uint32_t t_lane = static_cast<uint32_t>(quarter * 32) << 16;
    // pixel base pointer of local tile j (garbage pixels read pixel 0's in-range window)
    auto tile_img = [&](int j) -> const float * {
      const TcTile tt = tc_tile(a, n_fb, static_cast<int>(blockIdx.x) + j * static_cast<int>(gridDim.x));
      const int pp = tt.t * kM + row;
      const int y = pp / a.W, x = pp - y * a.W;
      const int pe = (y < a.Ho && x < a.Wo) ? pp : 0;
      return a.in + static_cast<size_t>(tt.n) * a.C * plane + pe;
    };
    auto load = [&](float (&v)[KS], int g) {
      const int j = g / a.n_kb, kb = g - j * a.n_kb;
      const float *__restrict__ img = tile_img(j);
      const int4 *ko = reinterpret_cast<const int4 *>(koff + kb * kKB + kpart * KS);
#pragma unroll
      for (int q = 0; q < KS / 4; ++q) {
        const int4 o = ko[q];
        v[4 * q + 0] = __ldg(img + o.x);
        v[4 * q + 1] = __ldg(img + o.y);
        v[4 * q + 2] = __ldg(img + o.z);
        v[4 * q + 3] = __ldg(img + o.w);
      }
    };
    auto put = [&](float (&v)[KS], int g) {
      const int s = g % NSA;
      if (g >= NSA) {
        mbar_wait(smem_u32(&empty_a[s]), static_cast<uint32_t>((g / NSA - 1) & 1));
        tc_fence_after();
      }
      const int kb = g % a.n_kb;
      if (kb == a.n_kb - 1) {  // padding k >= Kg: exact zeros
#pragma unroll
        for (int q = 0; q < KS; ++q)
          if (kb * kKB + kpart * KS + q >= a.Kg) v[q] = 0.f;
      }
      uint32_t hi[KS], lo[KS];
#pragma unroll
      for (int q = 0; q < KS; ++q) {
        const float h = tf32_hi_fast(v[q]);
        hi[q] = __float_as_uint(h);
        lo[q] = __float_as_uint(v[q] - h);
      }
      const uint32_t col = tmem + t_lane + Cfg::kAcc + s * 2 * kKB + kpart * KS;
      tmem_stv<KS>(col, hi);
      tmem_stv<KS>(col + kKB, lo);
      asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
      tc_fence_before();
      mbar_arrive(smem_u32(&full_a[s]));
    };
    // ring of D register buffers: blocks g+1 .. g+D-1 in flight while block g is split and stored
    float v[D][KS];
#pragma unroll
    for (int d = 0; d < D; ++d)
      if (d < n_blocks) load(v[d], d);
    for (int g0 = 0; g0 < n_blocks; g0 += D) {
#pragma unroll
      for (int d = 0; d < D; ++d) {
        const int g = g0 + d;
        if (g < n_blocks) {
          put(v[d], g);
          if (g + D < n_blocks) load(v[d], g + D);
        }
      }
    }
  } else if (warp < GW + 4) {
    // ---------------- epilogue: TMEM accumulator -> out[n][f][y][x] ----------------
    const int quarter = warp & 3;
    const int row = quarter * 32 + lane;
    const uint32_t t_lane = static_cast<uint32_t>(quarter * 32) << 16;
    const size_t PP = static_cast<size_t>(a.Ho) * a.Wo;
    for (int j = 0; j < my_tiles; ++j) {
      const int ab = j & 1;
      const TcTile tt = tc_tile(a, n_fb, static_cast<int>(blockIdx.x) + j * static_cast<int>(gridDim.x));
      const int pp = tt.t * kM + row;
      const int y = pp / a.W, x = pp - y * a.W;
      const bool valid = (y < a.Ho) && (x < a.Wo);
      float *__restrict__ obase = a.out + (static_cast<size_t>(tt.n) * a.F) * PP + (valid ? (y * a.Wo + x) : 0);
      const int f0 = tt.fblk * FN;
      mbar_wait(smem_u32(&acc_full[ab]), static_cast<uint32_t>((j >> 1) & 1));
      tc_fence_after();
#pragma unroll 1
      for (int c0 = 0; c0 < FN; c0 += 16) {
        float v[16];
        tmem_ld16(tmem + t_lane + ab * FN + c0, v);
        if (valid) {
#pragma unroll
          for (int q = 0; q < 16; ++q) {
            const int f = f0 + c0 + q;
            if (f < a.F) __stcs(obase + static_cast<size_t>(f) * PP, v[q]);
          }
        }
      }
      tc_fence_before();
      mbar_arrive(smem_u32(&acc_empty[ab]));
    }
  } else if (warp == Wp::kMma) {
    // ---------------- MMA issuer ----------------
    if (lane == 0) {
      constexpr uint32_t idesc = idesc_tf32(kM, FN);
      constexpr uint32_t lbo = (FN / 8) * 128;
      int g = 0;
      for (int j = 0; j < my_tiles; ++j) {
        const int ab = j & 1;
        if (j >= 2) {  // the epilogue of tile j-2 has drained this accumulator
          mbar_wait(smem_u32(&acc_empty[ab]), static_cast<uint32_t>(((j >> 1) - 1) & 1));
          tc_fence_after();
        }
        const uint32_t d = tmem + ab * FN;
        for (int kb = 0; kb < a.n_kb; ++kb, ++g) {
          const int sa = g % NSA, sb = b_resident ? kb : g % NSB;
          mbar_wait(smem_u32(&full_a[sa]), static_cast<uint32_t>((g / NSA) & 1));
          mbar_wait(smem_u32(&full_b[sb]), b_resident ? 0u : static_cast<uint32_t>((g / NSB) & 1));
          tc_fence_after();
          const uint32_t a_hi = tmem + Cfg::kAcc + sa * 2 * kKB, a_lo = a_hi + kKB;
          const uint32_t b_hi = sb_base + sb * Cfg::kBStage, b_lo = b_hi + Cfg::kBStage / 2;
#pragma unroll
          for (int kk = 0; kk < kKB / 8; ++kk) {
            const uint32_t bo = static_cast<uint32_t>(2 * kk * (FN / 8) * 128);
            const uint64_t dbh = umma_desc(b_hi + bo, lbo, 128), dbl = umma_desc(b_lo + bo, lbo, 128);
            const uint32_t acc0 = (kb > 0 || kk > 0) ? 1u : 0u;
            mma_tf32_ts(d, a_hi + 8 * kk, dbh, idesc, acc0);
            mma_tf32_ts(d, a_hi + 8 * kk, dbl, idesc, 1u);
            mma_tf32_ts(d, a_lo + 8 * kk, dbh, idesc, 1u);
          }
          mma_commit(smem_u32(&empty_a[sa]));
          if (!b_resident) mma_commit(smem_u32(&empty_b[sb]));
        }
        mma_commit(smem_u32(&acc_full[ab]));
      }
    }
  } else {
    // ---------------- B producer ----------------
    if (lane == 0 && b_resident) {  // every K block of the one filter block stays in shared memory
      for (int kb = 0; kb < a.n_kb; ++kb) {
        mbar_arrive_tx(smem_u32(&full_b[kb]), Cfg::kBStage);
        bulk_g2s(sb_base + kb * Cfg::kBStage, a.bs + static_cast<size_t>(kb) * (Cfg::kBStage / 4), Cfg::kBStage,
                 smem_u32(&full_b[kb]));
      }
    } else if (lane == 0) {
      int g = 0;
      for (int j = 0; j < my_tiles; ++j) {
        const TcTile tt = tc_tile(a, n_fb, static_cast<int>(blockIdx.x) + j * static_cast<int>(gridDim.x));
        const float *src = a.bs + static_cast<size_t>(tt.fblk) * a.n_kb * (Cfg::kBStage / 4);
        for (int kb = 0; kb < a.n_kb; ++kb, ++g) {
          const int sb = g % NSB;
          if (g >= NSB) mbar_wait(smem_u32(&empty_b[sb]), static_cast<uint32_t>((g / NSB - 1) & 1));
          mbar_arrive_tx(smem_u32(&full_b[sb]), Cfg::kBStage);
          bulk_g2s(sb_base + sb * Cfg::kBStage, src + static_cast<size_t>(kb) * (Cfg::kBStage / 4), Cfg::kBStage,
                   smem_u32(&full_b[sb]));
        }
      }
    }
  }
  tc_fence_before();
  __syncthreads();
  if (warp == Wp::kMma) {
    tc_fence_after();
    asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(Cfg::kAlloc));
  }
}

// Enable the dynamic shared memory a kernel instantiation may use, once per instantiation and DEVICE
// (cudaFuncSetAttribute acts on the current device only; a process may drive several GPUs).
struct MaxDyn {
  std::atomic<int> v[c2d::kMaxDevices] = {};
};
template <typename KernelT>
int enable_smem(KernelT kernel, MaxDyn &cache, int *max_dyn) {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= c2d::kMaxDevices) return CONV2D_ECUDA;
  const int known = cache.v[dev].load(std::memory_order_acquire);
  if (known > 0) {
    *max_dyn = known;
    return CONV2D_OK;
  }
  int optin = 0;
  cudaFuncAttributes fa;
  if (cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev) != cudaSuccess ||
      cudaFuncGetAttributes(&fa, kernel) != cudaSuccess) {
    (void)cudaGetLastError();
    return CONV2D_ECUDA;
  }
  const int avail = optin - static_cast<int>(fa.sharedSizeBytes);
  if (cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, avail) != cudaSuccess) {
    (void)cudaGetLastError();
    return CONV2D_ECUDA;
  }
  cache.v[dev].store(avail, std::memory_order_release);
  *max_dyn = avail;
  return CONV2D_OK;
}

// Split the filters into a stream-ordered scratch buffer from the library pool, run `body(bs, n_fb)`
// (the main kernel launch), free the scratch (stream-ordered).
template <int FN, typename Body>
int with_split_filters(const TcArgs &a, const float *filt, cudaStream_t stream, Body body) {
  const int n_fb = (a.F + FN - 1) / FN;
  const size_t bs_bytes = static_cast<size_t>(n_fb) * a.n_kb * (2u * FN * kKB * 4u);
  float *bs = nullptr;
  if (c2d::scratch_alloc(reinterpret_cast<void **>(&bs), bs_bytes, stream) != cudaSuccess) {
    (void)cudaGetLastError();
    return CONV2D_EALLOC;
  }
  int rc = CONV2D_OK;
  const long long split_elems = static_cast<long long>(n_fb) * a.n_kb * FN * kKB;
  const int split_blocks = static_cast<int>(split_elems / 256 < 1184 ? (split_elems + 255) / 256 : 1184);
  k_tc_split_filters<<<split_blocks, 256, 0, stream>>>(filt, a.F, a.Kg, FN, a.n_kb, n_fb, bs);
  if (cudaGetLastError() != cudaSuccess) rc = CONV2D_ECUDA;
  if (rc == CONV2D_OK) rc = body(bs, n_fb);
  if (cudaFreeAsync(bs, stream) != cudaSuccess && rc == CONV2D_OK) rc = CONV2D_ECUDA;
  return rc;
}

// one CTA per (pixel tile, filter block), two CTAs per SM
template <int FN, int D, int NBS = 0, int NACC = 1>
int launch_tc_d(TcArgs a, const float *filt, cudaStream_t stream) {
  using Cfg = TcCfg<FN, NBS, NACC>;
  auto kernel = k_conv2d_multi_tc4<FN, D, NBS, NACC>;
  const size_t smem = static_cast<size_t>(Cfg::NSB) * Cfg::kBStage + static_cast<size_t>(a.n_kb) * kKB * sizeof(int);
  static MaxDyn smem_cache;
  int max_dyn = 0;
  if (enable_smem(kernel, smem_cache, &max_dyn) != CONV2D_OK) return CONV2D_ECUDA;
  if (smem > static_cast<size_t>(max_dyn)) return CONV2D_ESHAPE;
  return with_split_filters<FN>(a, filt, stream, [&](const float *bs, int n_fb) {
    a.bs = bs;
    const dim3 grid(static_cast<unsigned>(static_cast<long long>(a.N) * a.tiles_per_img), static_cast<unsigned>(n_fb));
    kernel<<<grid, kThreads, smem, stream>>>(a);
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  });
}

// persistent: one CTA per SM over all (pixel tile, filter block) tiles
template <int FN, int D, int GW>
int launch_tc_p(TcArgs a, const float *filt, cudaStream_t stream) {
  using Cfg = TcPCfg<FN>;
  auto kernel = k_conv2d_multi_tc5<FN, D, GW>;
  const size_t smem = static_cast<size_t>(Cfg::NSB) * Cfg::kBStage + static_cast<size_t>(a.n_kb) * kKB * sizeof(int);
  static MaxDyn smem_cache;
  int max_dyn = 0;
  if (enable_smem(kernel, smem_cache, &max_dyn) != CONV2D_OK) return CONV2D_ECUDA;
  if (smem > static_cast<size_t>(max_dyn)) return CONV2D_ESHAPE;
  int dev = 0, n_sm = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || cudaDeviceGetAttribute(&n_sm, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess)
    return CONV2D_ECUDA;
  return with_split_filters<FN>(a, filt, stream, [&](const float *bs, int n_fb) {
    a.bs = bs;
    const long long tiles = static_cast<long long>(a.N) * a.tiles_per_img * n_fb;
    if (tiles > 2147483647LL) return CONV2D_ESHAPE;
    const int grid = static_cast<int>(tiles < n_sm ? tiles : n_sm);
    kernel<<<grid, TcPWarps<GW>::kThreads, smem, stream>>>(a, n_fb, static_cast<int>(tiles));
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  });
}

// Default: one CTA per (pixel tile, filter block), register ring depth 2, B ring of 2 stages. Tuning
// build only (c2d_debug_set_multi_variant): 41 / 42 = two accumulators (B ring 2 / 3), 23 / 24 = ring
// depth 3 / 4, 33 / 34 = a B ring of 3 / 4 stages, 50-55 = the persistent kernel (k_conv2d_multi_tc5).
template <int FN>
int launch_tc(const TcArgs &a, const float *filt, cudaStream_t stream) {
#ifdef C2D_TUNING
  const int mv = c2d::tuning_mvariant();
  if (mv == 41) return launch_tc_d<FN, 2, 2, 2>(a, filt, stream);
  if (mv == 42) return launch_tc_d<FN, 2, 3, 2>(a, filt, stream);
  if (mv == 23) return launch_tc_d<FN, 3>(a, filt, stream);
  if (mv == 24) return launch_tc_d<FN, 4>(a, filt, stream);
  if (mv == 33) return launch_tc_d<FN, 2, 3>(a, filt, stream);
  if (mv == 34) return launch_tc_d<FN, 2, 4>(a, filt, stream);
  if (mv == 50) return launch_tc_p<FN, 2, 8>(a, filt, stream);
  if (mv == 51) return launch_tc_p<FN, 3, 8>(a, filt, stream);
  if (mv == 52) return launch_tc_p<FN, 4, 8>(a, filt, stream);
  if (mv == 53) return launch_tc_p<FN, 2, 16>(a, filt, stream);
  if (mv == 54) return launch_tc_p<FN, 3, 16>(a, filt, stream);
  if (mv == 55) return launch_tc_p<FN, 4, 16>(a, filt, stream);
#endif
  return launch_tc_d<FN, 2, 2>(a, filt, stream);
}

}  // namespace c2d_tc

extern "C" int conv2d_multi_tc(const float *in, int N, int C, int H, int W, const float *filt, int F, int K,
                               float *out, void *stream) {
  using namespace c2d_tc;
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (K < 1) return CONV2D_ESHAPE;
  if (K > CONV2D_MAX_K) return CONV2D_EK;
  if (N < 1 || C < 1 || F < 1 || H < K || W < K) return CONV2D_ESHAPE;
  if ((reinterpret_cast<uintptr_t>(in) | reinterpret_cast<uintptr_t>(filt) | reinterpret_cast<uintptr_t>(out)) & 3u)
    return CONV2D_EALIGN;
  // 32-bit in-image offsets (one image's C planes) and a bounded im2col offset table
  if (static_cast<long long>(C) * H * W >= (1LL << 31) || static_cast<long long>(C) * K * K > (1 << 14))
    return CONV2D_ESHAPE;
  {  // the output may overlap neither the input nor the filters (as conv2d_multi)
    const uintptr_t o0 = reinterpret_cast<uintptr_t>(out);
    const uintptr_t o1 = o0 + static_cast<size_t>(N) * F * (H - K + 1) * (W - K + 1) * sizeof(float);
    const uintptr_t i0 = reinterpret_cast<uintptr_t>(in), i1 = i0 + static_cast<size_t>(N) * C * H * W * sizeof(float);
    const uintptr_t f0 = reinterpret_cast<uintptr_t>(filt), f1 = f0 + static_cast<size_t>(F) * C * K * K * sizeof(float);
    if ((o0 < i1 && i0 < o1) || (o0 < f1 && f0 < o1)) return CONV2D_EOVERLAP;
  }
  TcArgs a;
  a.in = in;
  a.bs = nullptr;
  a.out = out;
  a.N = N;
  a.C = C;
  a.H = H;
  a.W = W;
  a.F = F;
  a.K = K;
  a.Ho = H - K + 1;
  a.Wo = W - K + 1;
  a.Kg = C * K * K;
  a.n_kb = (a.Kg + kKB - 1) / kKB;
  a.tiles_per_img = static_cast<int>((static_cast<long long>(a.Ho) * W + kM - 1) / kM);
  if (static_cast<long long>(N) * a.tiles_per_img > 2147483647LL) return CONV2D_ESHAPE;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  // filter block FN = the smallest of 32/64/128 covering F (F > 128: several 128-filter blocks); a
  // smaller block when the larger one's shared memory (B ring + offset table) does not fit
  int rc = CONV2D_ESHAPE;
  if (F > 64) rc = launch_tc<128>(a, filt, s);
  if (rc == CONV2D_ESHAPE && F > 32) rc = launch_tc<64>(a, filt, s);
  if (rc == CONV2D_ESHAPE) rc = launch_tc<32>(a, filt, s);
  return rc;
}

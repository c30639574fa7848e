// conv2d_tc.cu -- tensor-core variant of the multi-channel convolution: the large-C
// case is a dense contraction, D[p][f] = sum_k A[p][k] * B[k][f] with p = (n, y, x) output pixels,
// f filters and k = (c, i, j), A[p][k] = in[n][c][y+i][x+j] (implicit im2col), B[k][f] = w[f][c][i][j].
// It runs on the 5th-generation tensor cores (tcgen05.mma kind::tf32, accumulator in TMEM) with the
// 3xTF32 split a = a_hi + a_lo (a_hi = tf32(a), a_lo = a - a_hi exact in fp32):
//     D = A_hi B_hi + A_hi B_lo + A_lo B_hi      (the dropped A_lo B_lo term is ~2^-22 |a||b|)
// which keeps each product within ~2^-21 relative, far inside the 1e-5 * sum|x||w| acceptance
// (DESIGN.md "Tensor-core variant"). A separate, measured variant, as BASELINE.json north_star asks.
//
// CTA = 128 threads, one 128-pixel x FN-filter output tile (FN <= 256, TMEM columns = FN), K in blocks
// of 32. Per K block every thread gathers its pixel's 32 im2col values (coalesced across the warp),
// splits them and writes A_hi / A_lo into shared memory in the canonical K-major no-swizzle UMMA layout
// (8-row x 16-byte core matrices); the filter block is split the same way into B_hi / B_lo. Two
// stages: while the tensor core runs block b, the threads stage block b+1. One elected thread issues
// 4 x 3 MMAs per block and commits them to the stage's mbarrier. The epilogue reads the accumulator
// with tcgen05.ld (each warp its 32 TMEM lanes) and stores NFHoWo rows (coalesced along pixels).
#include <cstdint>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"

namespace c2d_tc {

constexpr int kM = 128;     // pixels per tile (UMMA M)
constexpr int kKB = 32;     // k values per block (4 UMMA K=8 steps)
constexpr int kThreads = 256;  // 2 threads per pixel row: each stages 16 of a block's 32 k

__device__ __forceinline__ uint32_t smem_u32(const void *p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

__device__ __forceinline__ float tf32_hi(float a) {
  uint32_t r;
  asm("cvt.rna.tf32.f32 %0, %1;" : "=r"(r) : "f"(a));
  return __uint_as_float(r);
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

__device__ __forceinline__ void mma_tf32(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc,
                                         uint32_t accumulate) {
  asm volatile(
      "{\n\t.reg .pred p;\n\t"
      "setp.ne.b32 p, %4, 0;\n\t"
      "tcgen05.mma.cta_group::1.kind::tf32 [%0], %1, %2, %3, p;\n\t}\n" ::"r"(tmem_d),
      "l"(adesc), "l"(bdesc), "r"(idesc), "r"(accumulate));
}

__device__ __forceinline__ void mma_commit(uint32_t mbar) {
  asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(mbar)
               : "memory");
}

__device__ __forceinline__ void mbar_init(uint32_t mbar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(mbar), "r"(count) : "memory");
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

__device__ __forceinline__ void fence_async_smem() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }
__device__ __forceinline__ void tc_fence_before() { asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory"); }
__device__ __forceinline__ void tc_fence_after() { asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory"); }

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

struct TcArgs {
  const float *in;
  const float *filt;
  float *out;
  int N, C, H, W, F, K, Ho, Wo;
  long long P;   // N * Ho * Wo output pixels
  int Kg;        // C * K * K
  int n_kb;      // K blocks
  int f0;        // first filter of this launch's N tile
};

// stage bytes: A_hi, A_lo (128 x 32 fp32 each) + B_hi, B_lo (FN x 32 each)
template <int FN>
struct Stage {
  static constexpr uint32_t kA = kM * kKB * 4;   // 16 KiB
  static constexpr uint32_t kB = FN * kKB * 4;
  static constexpr uint32_t kBytes = 2 * kA + 2 * kB;
};

// element (row r, k) of a [rows x 32] K-major no-swizzle tile: core matrix (r/8, k/4) of 8 x 16 B
__device__ __forceinline__ uint32_t tile_off(int rows, int r, int k) {
  return static_cast<uint32_t>(((k >> 2) * (rows >> 3) + (r >> 3)) * 128 + (r & 7) * 16 + (k & 3) * 4);
}

template <int FN>
__global__ void __launch_bounds__(kThreads) k_conv2d_multi_tc3(const TcArgs a) {
  extern __shared__ __align__(1024) uint8_t smem[];  // [2 stages][A_hi A_lo B_hi B_lo] + int koff[Kg]
  __shared__ __align__(8) uint64_t mbar[2];
  __shared__ uint32_t tmem_base_s;
  constexpr uint32_t SB = Stage<FN>::kBytes;
  const uint32_t sbase = smem_u32(smem);
  const int tid = threadIdx.x;
  const int warp = tid >> 5;

  if (warp == 0) {  // TMEM accumulator: FN columns (power of two >= 32)
    asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(&tmem_base_s)),
                 "r"(FN));
    asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
  }
  if (tid == 0) {
    mbar_init(smem_u32(&mbar[0]), 1);
    mbar_init(smem_u32(&mbar[1]), 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  tc_fence_before();
  __syncthreads();
  tc_fence_after();
  const uint32_t tmem_d = tmem_base_s;

  // im2col offsets of every k = (c, i, j) relative to the pixel's (c=0, y, x) input element
  int *koff = reinterpret_cast<int *>(smem + 2 * SB);
  for (int k = tid; k < a.Kg; k += kThreads) {
    const int KK0 = a.K * a.K;
    const int c = k / KK0, ij = k - c * KK0;
    const int i = ij / a.K, j = ij - i * a.K;
    koff[k] = (c * a.H + i) * a.W + j;
  }
  __syncthreads();
  // this thread's pixel (row of A) and half of each K block
  const int row = tid & (kM - 1);
  const int khalf = tid / kM;  // 0 or 1: k in [16*khalf, 16*khalf+16) of each block
  const long long g = static_cast<long long>(blockIdx.x) * kM + row;
  const bool valid = g < a.P;
  const long long gg = valid ? g : a.P - 1;
  const int PP = a.Ho * a.Wo;
  const int n = static_cast<int>(gg / PP);
  const int p = static_cast<int>(gg % PP);
  const int y = p / a.Wo, x = p % a.Wo;
  const float *__restrict__ pix = a.in + (static_cast<size_t>(n) * a.C * a.H + y) * a.W + x;
  constexpr uint32_t idesc = idesc_tf32(kM, FN);

  // gather + split one K block into stage s
  auto stage_block = [&](int kb, int s) {
    const uint32_t st = sbase + s * SB;
    const int k0 = kb * kKB;
    // A: 16 values of this thread's im2col row (its half of the block), 4 at a time -> one 16-byte
    // store per (hi, lo); consecutive lanes = consecutive pixels, so each load is coalesced
#pragma unroll
    for (int q = 0; q < kKB / 8; ++q) {
      const int kq = 16 * khalf + 4 * q;
      float hi[4], lo[4];
#pragma unroll
      for (int t = 0; t < 4; ++t) {
        const int k = k0 + kq + t;
        const float v = (k < a.Kg) ? __ldg(pix + koff[k]) : 0.f;
        hi[t] = tf32_hi(v);
        lo[t] = v - hi[t];
      }
      const uint32_t off = tile_off(kM, row, kq);
      asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(st + off), "f"(hi[0]), "f"(hi[1]), "f"(hi[2]),
                   "f"(hi[3]) : "memory");
      asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(st + Stage<FN>::kA + off), "f"(lo[0]),
                   "f"(lo[1]), "f"(lo[2]), "f"(lo[3]) : "memory");
    }
    // B: FN filter rows x 32 k (contiguous in FCKK), 4 at a time
    for (int e = tid; e < FN * (kKB / 4); e += kThreads) {
      const int f = e / (kKB / 4), q = e % (kKB / 4);
      const int fg = a.f0 + f;
      float hi[4], lo[4];
#pragma unroll
      for (int t = 0; t < 4; ++t) {
        const int k = k0 + 4 * q + t;
        const float v = (fg < a.F && k < a.Kg) ? __ldg(a.filt + static_cast<size_t>(fg) * a.Kg + k) : 0.f;
        hi[t] = tf32_hi(v);
        lo[t] = v - hi[t];
      }
      const uint32_t off = tile_off(FN, f, 4 * q);
      asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(st + 2 * Stage<FN>::kA + off), "f"(hi[0]),
                   "f"(hi[1]), "f"(hi[2]), "f"(hi[3]) : "memory");
      asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(st + 2 * Stage<FN>::kA + Stage<FN>::kB + off),
                   "f"(lo[0]), "f"(lo[1]), "f"(lo[2]), "f"(lo[3]) : "memory");
    }
    fence_async_smem();  // generic-proxy smem writes -> visible to the tensor core (async proxy)
  };

  auto issue_block = [&](int kb, int s) {
    const uint32_t st = sbase + s * SB;
    const uint32_t a_hi = st, a_lo = st + Stage<FN>::kA;
    const uint32_t b_hi = st + 2 * Stage<FN>::kA, b_lo = b_hi + Stage<FN>::kB;
#pragma unroll
    for (int kk = 0; kk < kKB / 8; ++kk) {
      // K = 8 tf32 = two 16-byte chunks: chunk (2kk) and (2kk+1) of the tile
      const uint32_t ao = static_cast<uint32_t>(2 * kk * (kM / 8) * 128);
      const uint32_t bo = static_cast<uint32_t>(2 * kk * (FN / 8) * 128);
      const uint32_t a_lbo = (kM / 8) * 128, b_lbo = (FN / 8) * 128;
      const uint64_t dah = umma_desc(a_hi + ao, a_lbo, 128), dal = umma_desc(a_lo + ao, a_lbo, 128);
      const uint64_t dbh = umma_desc(b_hi + bo, b_lbo, 128), dbl = umma_desc(b_lo + bo, b_lbo, 128);
      const uint32_t acc0 = (kb > 0 || kk > 0) ? 1u : 0u;
      mma_tf32(tmem_d, dah, dbh, idesc, acc0);
      mma_tf32(tmem_d, dah, dbl, idesc, 1u);
      mma_tf32(tmem_d, dal, dbh, idesc, 1u);
    }
    mma_commit(smem_u32(&mbar[s]));
  };

  // two-stage pipeline: stage kb+1 while the tensor core runs kb
  uint32_t phase[2] = {0u, 0u};
  stage_block(0, 0);
  __syncthreads();
  for (int kb = 0; kb < a.n_kb; ++kb) {
    const int s = kb & 1;
    if (tid == 0) {
      tc_fence_after();
      issue_block(kb, s);
    }
    if (kb + 1 < a.n_kb) {
      const int s2 = s ^ 1;
      if (kb >= 1) {  // stage s2 was consumed by the MMAs of block kb-1
        mbar_wait(smem_u32(&mbar[s2]), phase[s2]);
        phase[s2] ^= 1u;
      }
      stage_block(kb + 1, s2);
    }
    __syncthreads();
  }
  // the last block's commit tracks every MMA issued before it: its completion means D is final
  // (every earlier commit of that stage was waited on above, so phase[] is current)
  {
    const int s_last = (a.n_kb - 1) & 1;
    mbar_wait(smem_u32(&mbar[s_last]), phase[s_last]);
  }
  tc_fence_after();

  // epilogue: TMEM -> registers -> out[n][f][p]. Warp w may only access TMEM lanes 32(w%4)..+31, so
  // warps w and w+4 split the accumulator columns of the same 32 pixels.
  const uint32_t lane_base = static_cast<uint32_t>((warp & 3) * 32) << 16;
#pragma unroll 1
  for (int c0 = 16 * khalf; c0 < FN; c0 += 32) {
    float v[16];
    tmem_ld16(tmem_d + lane_base + c0, v);
    if (valid) {
#pragma unroll
      for (int t = 0; t < 16; ++t) {
        const int f = a.f0 + c0 + t;
        if (f < a.F) a.out[(static_cast<size_t>(n) * a.F + f) * PP + p] = v[t];
      }
    }
  }
  tc_fence_before();
  __syncthreads();
  if (warp == 0)
    asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem_d), "r"(FN));
}

template <int FN>
int launch_tc(const TcArgs &a0, cudaStream_t stream) {
  auto kernel = k_conv2d_multi_tc3<FN>;
  const size_t smem = 2 * Stage<FN>::kBytes + static_cast<size_t>(a0.Kg) * sizeof(int);
  static int max_dyn = 0;  // dynamic shared memory enabled for this instantiation
  if (max_dyn == 0) {
    int dev = 0, optin = 0;
    cudaFuncAttributes fa;
    if (cudaGetDevice(&dev) != cudaSuccess ||
        cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev) != cudaSuccess ||
        cudaFuncGetAttributes(&fa, kernel) != cudaSuccess) {
      (void)cudaGetLastError();
      return CONV2D_ECUDA;
    }
    const int avail = optin - static_cast<int>(fa.sharedSizeBytes);
    if (cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, avail) != cudaSuccess) {
      (void)cudaGetLastError();
      return CONV2D_ECUDA;
    }
    max_dyn = avail;
  }
  if (smem > static_cast<size_t>(max_dyn)) return CONV2D_ESHAPE;
  TcArgs a = a0;
  const long long blocks = (a.P + kM - 1) / kM;
  for (int f0 = 0; f0 < a.F; f0 += FN) {
    a.f0 = f0;
    kernel<<<static_cast<unsigned>(blocks), kThreads, smem, stream>>>(a);
    if (cudaGetLastError() != cudaSuccess) return CONV2D_ECUDA;
  }
  return CONV2D_OK;
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
  TcArgs a;
  a.in = in;
  a.filt = filt;
  a.out = out;
  a.N = N;
  a.C = C;
  a.H = H;
  a.W = W;
  a.F = F;
  a.K = K;
  a.Ho = H - K + 1;
  a.Wo = W - K + 1;
  a.P = static_cast<long long>(N) * a.Ho * a.Wo;
  a.Kg = C * K * K;
  a.n_kb = (a.Kg + kKB - 1) / kKB;
  a.f0 = 0;
  const double px = static_cast<double>(a.P);
  if (px / kM > 2147483647.0) return CONV2D_ESHAPE;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  if (F <= 32) return launch_tc<32>(a, s);
  if (F <= 64) return launch_tc<64>(a, s);
  if (F <= 128) return launch_tc<128>(a, s);
  return launch_tc<256>(a, s);
}

// conv2d_pad.cu -- boundary and semantic variants of the single-channel call:
// 'same' output size with zero or replicate padding, and true (flipped-filter) convolution.
//
// Both reduce to the valid-mode, stride-1 cross-correlation the paper's kernels compute (PAPER.md
// P:83-85; R1/R2): true convolution is cross-correlation with the filter rotated
// by 180 degrees, and 'same' is the valid result on the image padded by K-1 rows and columns
// (top/left (K-1)/2, bottom/right K-1-(K-1)/2, the convention of torch.nn.functional.conv2d
// padding='same'). The rotation and the padding are pure data movement done by two small kernels
// into the library's stream-ordered scratch pool; the padded image gets a 16-byte row pitch so the
// convolution takes the vectorised row-fetch path; then the same per-K kernels as conv2d_single run
// on it. Results are therefore bitwise equal to conv2d_single on the padded image / rotated filter.
// (In-kernel padding would save the extra pass over the image -- ~2x traffic at HBM-bound K = 3 and
// a few percent at FMA-bound K -- at the cost of another edge path through the hot kernels.)
#include <cstdint>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"
#include "common.h"

namespace {

using namespace c2d;

// P[r][c] (r < Hp, c < P4*4) from in (H x W): padded column c maps to input column c - pl, row r to
// input row r - pt; out-of-range entries are 0 (ZERO) or the nearest edge element (REPLICATE);
// columns >= Wt (the pitch slack) are 0.
__global__ void k_pad_image(const float *__restrict__ in, int H, int W, float *__restrict__ P, int Hp, int Wt,
                            long long P4, int pt, int pl, int replicate) {
  const long long total = static_cast<long long>(Hp) * P4;
  for (long long q = static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x; q < total;
       q += static_cast<long long>(gridDim.x) * blockDim.x) {
    const int r = static_cast<int>(q / P4);
    const int c0 = static_cast<int>(q % P4) * 4;
    int ri = r - pt;
    const bool row_in = ri >= 0 && ri < H;
    if (replicate) ri = min(max(ri, 0), H - 1);
    float v[4];
#pragma unroll
    for (int t = 0; t < 4; ++t) {
      const int c = c0 + t;
      int ci = c - pl;
      const bool col_in = ci >= 0 && ci < W;
      if (replicate) ci = min(max(ci, 0), W - 1);
      const bool take = c < Wt && (replicate || (row_in && col_in));
      v[t] = take ? __ldg(in + static_cast<long long>(ri) * W + ci) : 0.f;
    }
    reinterpret_cast<float4 *>(P)[q] = make_float4(v[0], v[1], v[2], v[3]);
  }
}

// fo[i][j] = f[K-1-i][K-1-j] (rotation by 180 degrees: convolution -> cross-correlation)
__global__ void k_rotate_filter(const float *__restrict__ f, int K, float *__restrict__ fo) {
  for (int t = threadIdx.x; t < K * K; t += blockDim.x) fo[t] = f[K * K - 1 - t];
}

bool overlap(const void *a, size_t abytes, const void *b, size_t bbytes) {
  const uintptr_t a0 = reinterpret_cast<uintptr_t>(a), b0 = reinterpret_cast<uintptr_t>(b);
  return a0 < b0 + bbytes && b0 < a0 + abytes;
}

int device_info(DevInfo *out) {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess) return CONV2D_ECUDA;
  if (cudaDeviceGetAttribute(&out->num_sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess ||
      cudaDeviceGetAttribute(&out->smem_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev) != cudaSuccess)
    return CONV2D_ECUDA;
  return CONV2D_OK;
}

}  // namespace

extern "C" int conv2d_single_pad(const float *in, int H, int W, const float *filt, int K, int mode, float *out,
                                 void *stream) {
  if ((mode & ~(CONV2D_PAD_MASK | CONV2D_FLIP)) != 0 || (mode & CONV2D_PAD_MASK) == CONV2D_PAD_MASK)
    return CONV2D_ESHAPE;
  const int pad = mode & CONV2D_PAD_MASK;
  const bool flip = (mode & CONV2D_FLIP) != 0;
  if (!pad && !flip) return conv2d_single_ex(in, H, W, filt, K, out, stream, 0);
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (K < 1) return CONV2D_ESHAPE;
  if (K > CONV2D_MAX_K) return CONV2D_EK;
  if (H < 1 || W < 1 || (!pad && (H < K || W < K))) return CONV2D_ESHAPE;
  if ((reinterpret_cast<uintptr_t>(in) | reinterpret_cast<uintptr_t>(filt) | reinterpret_cast<uintptr_t>(out)) & 3u)
    return CONV2D_EALIGN;
  const long long Ht = pad ? static_cast<long long>(H) + K - 1 : H;
  const long long Wt = pad ? static_cast<long long>(W) + K - 1 : W;
  if (Ht > 0x7fffffffLL || Wt > 0x7fffffffLL) return CONV2D_ESHAPE;
  const long long Ho = Ht - K + 1, Wo = Wt - K + 1;
  const size_t in_b = static_cast<size_t>(H) * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(Ho) * Wo * sizeof(float);
  const size_t f_b = static_cast<size_t>(K) * K * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(filt, f_b, out, out_b)) return CONV2D_EOVERLAP;
  DevInfo dev;
  if (device_info(&dev)) return CONV2D_ECUDA;
  cudaStream_t s = static_cast<cudaStream_t>(stream);

  const float *f_use = filt;
  float *f_rot = nullptr;
  if (flip) {
    if (scratch_alloc(reinterpret_cast<void **>(&f_rot), f_b, s) != cudaSuccess) return CONV2D_EALLOC;
    k_rotate_filter<<<1, 256, 0, s>>>(filt, K, f_rot);
    if (cudaGetLastError() != cudaSuccess) {
      cudaFreeAsync(f_rot, s);
      return CONV2D_ECUDA;
    }
    f_use = f_rot;
  }
  const float *src = in;
  long long pitch = W;
  float *padded = nullptr;
  if (pad) {
    pitch = (Wt + 3) / 4 * 4;  // 16-byte rows: the vectorised row fetch
    const size_t p_b = static_cast<size_t>(Ht) * pitch * sizeof(float);
    if (scratch_alloc(reinterpret_cast<void **>(&padded), p_b, s) != cudaSuccess) {
      if (f_rot) cudaFreeAsync(f_rot, s);
      return CONV2D_EALLOC;
    }
    const long long quads = Ht * (pitch / 4);
    long long blocks = (quads + 255) / 256;
    const long long cap = static_cast<long long>(dev.num_sms) * 8;
    if (blocks > cap) blocks = cap;
    k_pad_image<<<static_cast<unsigned>(blocks), 256, 0, s>>>(in, H, W, padded, static_cast<int>(Ht),
                                                              static_cast<int>(Wt), pitch / 4, (K - 1) / 2,
                                                              (K - 1) / 2, pad == CONV2D_PAD_REPLICATE ? 1 : 0);
    if (cudaGetLastError() != cudaSuccess) {
      cudaFreeAsync(padded, s);
      if (f_rot) cudaFreeAsync(f_rot, s);
      return CONV2D_ECUDA;
    }
    src = padded;
  }
  const int Hi = static_cast<int>(Ht), Wi = static_cast<int>(Wt);
  int rc;
#define C2D_CALL_PAD(KK) rc = single_entry<KK>(src, Hi, Wi, f_use, out, s, 0, dev, src, Hi, pitch); break;
  switch (K) {
    case 1: C2D_CALL_PAD(1)
    case 2: C2D_CALL_PAD(2)
    case 3: C2D_CALL_PAD(3)
    case 4: C2D_CALL_PAD(4)
    case 5: C2D_CALL_PAD(5)
    case 6: C2D_CALL_PAD(6)
    case 7: C2D_CALL_PAD(7)
    case 8: C2D_CALL_PAD(8)
    case 9: C2D_CALL_PAD(9)
    case 10: C2D_CALL_PAD(10)
    case 11: C2D_CALL_PAD(11)
    case 12: C2D_CALL_PAD(12)
    case 13: C2D_CALL_PAD(13)
    case 14: C2D_CALL_PAD(14)
    default: C2D_CALL_PAD(15)
  }
#undef C2D_CALL_PAD
  // scratch returns to the pool once the convolution (ordered before on s) has read it
  if (padded) cudaFreeAsync(padded, s);
  if (f_rot) cudaFreeAsync(f_rot, s);
  return rc;
}

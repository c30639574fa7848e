// conv2d_capi.cu -- the C ABI declared in include/conv2d.h: argument validation and per-K dispatch
// to the launch units (inst_kNN.cu), the Fig. 1a baseline kernel, error strings.
#include <atomic>
#include <cstdint>
#include <mutex>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"
#include "common.h"

namespace c2d {

#ifdef C2D_TUNING
std::atomic<int> g_variant{0};
std::atomic<int> g_min_band{0};
std::atomic<int> g_mvariant{0};
#endif

// ------------------------------------------------------------------------------------------------
// Baseline: PAPER.md Fig. 1a direct convolution, one thread per output, K*K loads per thread
// ------------------------------------------------------------------------------------------------
__global__ void __launch_bounds__(256) k_conv2d_direct(const float *__restrict__ in, int W, const float *__restrict__ filt,
                                                       int K, float *__restrict__ out, int Ho, int Wo) {
  const long long idx = static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x;
  if (idx >= static_cast<long long>(Ho) * Wo) return;
  const int y = static_cast<int>(idx / Wo), x = static_cast<int>(idx % Wo);
  float s = 0.f;
  for (int i = 0; i < K; ++i)
    for (int j = 0; j < K; ++j) s = fmaf(in[static_cast<size_t>(y + i) * W + x + j], __ldg(filt + i * K + j), s);
  out[idx] = s;
}

// ------------------------------------------------------------------------------------------------
// library-owned stream-ordered scratch pool, one per device
// ------------------------------------------------------------------------------------------------
namespace {
constexpr int kPoolDevices = 64;
std::mutex g_pool_mu;
cudaMemPool_t g_pool[kPoolDevices] = {};
}  // namespace

cudaError_t scratch_alloc(void **p, size_t bytes, cudaStream_t stream) {
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  if (dev < 0 || dev >= kPoolDevices) return cudaErrorInvalidDevice;
  cudaMemPool_t pool;
  {
    std::lock_guard<std::mutex> lk(g_pool_mu);
    if (!g_pool[dev]) {
      cudaMemPoolProps props = {};
      props.allocType = cudaMemAllocationTypePinned;
      props.handleTypes = cudaMemHandleTypeNone;
      props.location.type = cudaMemLocationTypeDevice;
      props.location.id = dev;
      cudaMemPool_t np;
      if ((e = cudaMemPoolCreate(&np, &props)) != cudaSuccess) return e;
      uint64_t keep = ~0ull;
      if ((e = cudaMemPoolSetAttribute(np, cudaMemPoolAttrReleaseThreshold, &keep)) != cudaSuccess) return e;
      g_pool[dev] = np;
    }
    pool = g_pool[dev];
  }
  return cudaMallocFromPoolAsync(p, bytes, pool, stream);
}

cudaError_t scratch_trim() {
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  if (dev < 0 || dev >= kPoolDevices) return cudaErrorInvalidDevice;
  std::lock_guard<std::mutex> lk(g_pool_mu);
  return g_pool[dev] ? cudaMemPoolTrimTo(g_pool[dev], 0) : cudaSuccess;
}

}  // namespace c2d

namespace {

using namespace c2d;

DevInfo g_dev[kMaxDevices];
std::once_flag g_dev_once[kMaxDevices];

int current_device_info(DevInfo *out) {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= kMaxDevices) return CONV2D_ECUDA;
  std::call_once(g_dev_once[dev], [dev] {
    g_dev[dev].id = dev;
    cudaDeviceGetAttribute(&g_dev[dev].num_sms, cudaDevAttrMultiProcessorCount, dev);
    cudaDeviceGetAttribute(&g_dev[dev].smem_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
  });
  *out = g_dev[dev];
  return out->num_sms > 0 ? CONV2D_OK : CONV2D_ECUDA;
}

bool aligned4(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 3u) == 0; }

bool overlap(const void *a, size_t abytes, const void *b, size_t bbytes) {
  const uintptr_t a0 = reinterpret_cast<uintptr_t>(a), b0 = reinterpret_cast<uintptr_t>(b);
  return a0 < b0 + bbytes && b0 < a0 + abytes;
}

#define C2D_K_SWITCH(K, CALL) \
  switch (K) {                \
    case 1: return CALL(1);   \
    case 2: return CALL(2);   \
    case 3: return CALL(3);   \
    case 4: return CALL(4);   \
    case 5: return CALL(5);   \
    case 6: return CALL(6);   \
    case 7: return CALL(7);   \
    case 8: return CALL(8);   \
    case 9: return CALL(9);   \
    case 10: return CALL(10); \
    case 11: return CALL(11); \
    case 12: return CALL(12); \
    case 13: return CALL(13); \
    case 14: return CALL(14); \
    case 15: return CALL(15); \
    default: return CONV2D_EK; \
  }

int check_k(int K) {
  if (K < 1) return CONV2D_ESHAPE;
  if (K > CONV2D_MAX_K) return CONV2D_EK;
  return CONV2D_OK;
}

// Validation shared by the one-image and the batched call (N images of H x W, dense, back to back).
int single_batch_impl(const float *in, int N, int H, int W, const float *filt, int K, float *out, void *stream,
                      int band_h) {
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (int e = check_k(K)) return e;
  if (N < 1 || H < K || W < K) return CONV2D_ESHAPE;
  if (!aligned4(in) || !aligned4(filt) || !aligned4(out)) return CONV2D_EALIGN;
  const double in_n = static_cast<double>(N) * H * W;
  if (in_n > 4.0e18 || static_cast<double>(N) * (H - K + 1) * (W - K + 1) * 1.0 > 4.0e18) return CONV2D_ESHAPE;
  const size_t in_b = static_cast<size_t>(N) * H * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(N) * (H - K + 1) * (W - K + 1) * sizeof(float);
  const size_t f_b = static_cast<size_t>(K) * K * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(filt, f_b, out, out_b)) return CONV2D_EOVERLAP;
  DevInfo dev;
  if (current_device_info(&dev)) return CONV2D_ECUDA;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
#define C2D_CALL_SINGLE(KK) single_entry<KK>(in, N, H, W, filt, out, s, band_h, dev, in, H, W, W - KK + 1)
  C2D_K_SWITCH(K, C2D_CALL_SINGLE)
#undef C2D_CALL_SINGLE
}

}  // namespace

extern "C" {

int conv2d_single_ex(const float *in, int H, int W, const float *filt, int K, float *out, void *stream,
                     int band_h) {
  return single_batch_impl(in, 1, H, W, filt, K, out, stream, band_h);
}

int conv2d_single_batch(const float *in, int N, int H, int W, const float *filt, int K, float *out, void *stream) {
  return single_batch_impl(in, N, H, W, filt, K, out, stream, 0);
}

int conv2d_single_rect(const float *in, int H, int W, const float *filt, int FH, int FW, float *out,
                       void *stream) {
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (FH < 1 || FW < 1) return CONV2D_ESHAPE;
  if (FH > CONV2D_MAX_K || FW > CONV2D_MAX_K) return CONV2D_EK;
  if (H < FH || W < FW) return CONV2D_ESHAPE;
  if (!aligned4(in) || !aligned4(filt) || !aligned4(out)) return CONV2D_EALIGN;
  const size_t in_b = static_cast<size_t>(H) * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(H - FH + 1) * (W - FW + 1) * sizeof(float);
  const size_t f_b = static_cast<size_t>(FH) * FW * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(filt, f_b, out, out_b)) return CONV2D_EOVERLAP;
  if (FH == FW) return single_batch_impl(in, 1, H, W, filt, FH, out, stream, 0);  // square: conv2d_single
  DevInfo dev;
  if (current_device_info(&dev)) return CONV2D_ECUDA;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
#define C2D_CALL_RECT(KK) rect_entry<KK>(in, H, W, filt, FW, out, s, dev)
  C2D_K_SWITCH(FH, C2D_CALL_RECT)
#undef C2D_CALL_RECT
}

int conv2d_single_halo(const float *in, int H, int W, const float *halo, int halo_rows, const float *filt, int K,
                       float *out, void *stream) {
  if (halo_rows < 0) return CONV2D_ESHAPE;
  if (halo_rows == 0) return conv2d_single_ex(in, H, W, filt, K, out, stream, 0);
  if (!in || !halo || !filt || !out) return CONV2D_ENULL;
  if (int e = check_k(K)) return e;
  if (H < 1 || W < K) return CONV2D_ESHAPE;
  const long long Ht = static_cast<long long>(H) + halo_rows;
  if (Ht < K || Ht > 0x7fffffffLL) return CONV2D_ESHAPE;
  if (!aligned4(in) || !aligned4(halo) || !aligned4(filt) || !aligned4(out)) return CONV2D_EALIGN;
  const size_t in_b = static_cast<size_t>(H) * W * sizeof(float);
  const size_t halo_b = static_cast<size_t>(halo_rows) * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(Ht - K + 1) * (W - K + 1) * sizeof(float);
  const size_t f_b = static_cast<size_t>(K) * K * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(halo, halo_b, out, out_b) || overlap(filt, f_b, out, out_b))
    return CONV2D_EOVERLAP;
  DevInfo dev;
  if (current_device_info(&dev)) return CONV2D_ECUDA;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  const int Hi = static_cast<int>(Ht);
#define C2D_CALL_HALO(KK) single_entry<KK>(in, 1, Hi, W, filt, out, s, 0, dev, halo, H, W, W - KK + 1)
  C2D_K_SWITCH(K, C2D_CALL_HALO)
#undef C2D_CALL_HALO
}

int conv2d_single(const float *in, int H, int W, const float *filt, int K, float *out, void *stream) {
  return conv2d_single_ex(in, H, W, filt, K, out, stream, 0);
}

int conv2d_multi_ex(const float *in, int N, int C, int H, int W, const float *filt, int F, int K, float *out,
                    void *stream, int band_h) {
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (int e = check_k(K)) return e;
  if (N < 1 || C < 1 || F < 1 || H < K || W < K) return CONV2D_ESHAPE;
  if (!aligned4(in) || !aligned4(filt) || !aligned4(out)) return CONV2D_EALIGN;
  // element counts must fit comfortably in 64 bits
  const double in_n = static_cast<double>(N) * C * H * W;
  const double out_n = static_cast<double>(N) * F * (H - K + 1) * (W - K + 1);
  if (in_n > 4.0e18 || out_n > 4.0e18) return CONV2D_ESHAPE;
  const size_t in_b = static_cast<size_t>(N) * C * H * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(N) * F * (H - K + 1) * (W - K + 1) * sizeof(float);
  const size_t f_b = static_cast<size_t>(F) * C * K * K * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(filt, f_b, out, out_b)) return CONV2D_EOVERLAP;
  DevInfo dev;
  if (current_device_info(&dev)) return CONV2D_ECUDA;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
#define C2D_CALL_MULTI(KK) multi_entry<KK>(in, N, C, H, W, filt, F, out, s, band_h, dev)
  C2D_K_SWITCH(K, C2D_CALL_MULTI)
#undef C2D_CALL_MULTI
}

int conv2d_multi(const float *in, int N, int C, int H, int W, const float *filt, int F, int K, float *out,
                 void *stream) {
  return conv2d_multi_ex(in, N, C, H, W, filt, F, K, out, stream, 0);
}

int conv2d_single_direct(const float *in, int H, int W, const float *filt, int K, float *out, void *stream) {
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (int e = check_k(K)) return e;
  if (H < K || W < K) return CONV2D_ESHAPE;
  if (!aligned4(in) || !aligned4(filt) || !aligned4(out)) return CONV2D_EALIGN;
  const int Ho = H - K + 1, Wo = W - K + 1;
  const size_t in_b = static_cast<size_t>(H) * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(Ho) * Wo * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(filt, static_cast<size_t>(K) * K * 4, out, out_b))
    return CONV2D_EOVERLAP;
  const long long n = static_cast<long long>(Ho) * Wo;
  const long long blocks = (n + 255) / 256;
  if (blocks > 0x7fffffffLL) return CONV2D_ESHAPE;
  k_conv2d_direct<<<static_cast<unsigned>(blocks), 256, 0, static_cast<cudaStream_t>(stream)>>>(in, W, filt, K, out,
                                                                                                  Ho, Wo);
  return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
}

const char *conv2d_strerror(int code) {
  switch (code) {
    case CONV2D_OK: return "ok";
    case CONV2D_ENULL: return "a tensor pointer is NULL";
    case CONV2D_ESHAPE: return "bad shape (H<K, W<K, N/C/F<1, K<1, size overflow, or filters too large)";
    case CONV2D_EK: return "unsupported K (> 15)";
    case CONV2D_EOVERLAP: return "output overlaps input or filter";
    case CONV2D_ECUDA: return "CUDA launch error";
    case CONV2D_EALIGN: return "a tensor pointer is not 4-byte aligned";
    case CONV2D_EALLOC: return "device memory for a host-buffer call could not be allocated";
    default: return "unknown error code";
  }
}

int conv2d_version(void) { return 103; }

int conv2d_release_scratch(void) { return scratch_trim() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA; }

#ifdef C2D_TUNING
// Tuning build only (libconv2d_tune.so; not part of include/conv2d.h): force a kernel variant for
// tuning tools and the variant tests (0 = default).
int c2d_debug_set_variant(int v) { return g_variant.exchange(v); }

// multi-channel variant (0 = default; 1/2 FB wide/narrow segments, 3/4 half FB, 5/6 two column chunks,
// 7 8-lane segments, 9 = round-1 kernel)
int c2d_debug_set_multi_variant(int v) { return g_mvariant.exchange(v); }

// minimum band height override (0 = default)
int c2d_debug_set_min_band(int v) { return g_min_band.exchange(v); }
#endif

}  // extern "C"

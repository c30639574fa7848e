// conv2d_capi.cu -- the C ABI declared in include/conv2d.h: argument validation, launch geometry
// (band height, F-block), per-K template dispatch, launch on the caller's stream.
#include <atomic>
#include <cstdint>
#include <cstring>
#include <mutex>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"
#include "conv2d_kernels.cuh"

namespace {

using namespace c2d;

constexpr int kMaxDevices = 64;

struct DevInfo {
  int num_sms = 0;
  int smem_optin = 0;
};

DevInfo g_dev[kMaxDevices];
std::once_flag g_dev_once[kMaxDevices];

int current_device_info(DevInfo *out) {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= kMaxDevices) return CONV2D_ECUDA;
  std::call_once(g_dev_once[dev], [dev] {
    cudaDeviceGetAttribute(&g_dev[dev].num_sms, cudaDevAttrMultiProcessorCount, dev);
    cudaDeviceGetAttribute(&g_dev[dev].smem_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
  });
  *out = g_dev[dev];
  return out->num_sms > 0 ? CONV2D_OK : CONV2D_ECUDA;
}

bool aligned4(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 3u) == 0; }
bool aligned16(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 15u) == 0; }

bool overlap(const void *a, size_t abytes, const void *b, size_t bbytes) {
  const uintptr_t a0 = reinterpret_cast<uintptr_t>(a), b0 = reinterpret_cast<uintptr_t>(b);
  return a0 < b0 + bbytes && b0 < a0 + abytes;
}

int ceil_div(long long a, long long b) { return static_cast<int>((a + b - 1) / b); }

// Occupancy (CTAs per SM) of a kernel instantiation, cached per instantiation (devices of one box
// are identical B200s).
template <typename KernelT>
int cta_occupancy(KernelT kernel, size_t dyn_smem, std::atomic<int> &cache, int cta_warps = kCtaWarps) {
  int v = cache.load(std::memory_order_relaxed);
  if (v > 0) return v;
  int blocks = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, kernel, cta_warps * kWarp, dyn_smem) != cudaSuccess ||
      blocks < 1)
    blocks = 1;
  cache.store(blocks, std::memory_order_relaxed);
  return blocks;
}

// ------------------------------------------------------------------------------------------------
// single channel
// ------------------------------------------------------------------------------------------------
// Variant override for tuning tools (c2d_debug_set_variant; 0 = the tuned default):
//   1: filter in shared memory, U=1 (4 warps/CTA)     2: shared memory, U=2
//   3: filter in a __constant__ slot, U=1 (1 warp/CTA) 4: __constant__ slot, U=2
std::atomic<int> g_variant{0};
std::atomic<int> g_min_band{0};  // tuning override of the minimum band height (0 = per-K default)

// Constant-bank filter slots, per device: slot K holds the filter of the last call with this K. A
// call waits (stream-ordered) for the event recorded behind the previous kernel that read the slot
// before overwriting it, so calls on different streams never see each other's filter; calls with
// the same K on different streams are serialised by that wait, calls on one stream cost nothing.
struct ConstRing {
  std::mutex mu;
  bool init = false;
  float *base = nullptr;  // device address of c_filt
  cudaEvent_t ev[kConstSlots];
};
ConstRing g_cring[kMaxDevices];

template <typename LaunchFn>
int with_const_filter(const float *filt, int K, int KP, cudaStream_t stream, LaunchFn launch) {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= kMaxDevices) return CONV2D_ECUDA;
  ConstRing &ring = g_cring[dev];
  std::lock_guard<std::mutex> lk(ring.mu);
  if (!ring.init) {
    void *p = nullptr;
    if (cudaGetSymbolAddress(&p, c_filt) != cudaSuccess) return CONV2D_ECUDA;
    ring.base = static_cast<float *>(p);
    for (int i = 0; i < kConstSlots; ++i)
      if (cudaEventCreateWithFlags(&ring.ev[i], cudaEventDisableTiming) != cudaSuccess) return CONV2D_ECUDA;
    ring.init = true;
  }
  const int slot = K;
  if (cudaStreamWaitEvent(stream, ring.ev[slot], 0) != cudaSuccess) return CONV2D_ECUDA;
  // K rows of K floats -> K rows of KP floats (16-byte aligned rows for LDCU.128)
  if (cudaMemcpy2DAsync(ring.base + static_cast<size_t>(slot) * kConstSlotFloats, KP * sizeof(float), filt,
                        K * sizeof(float), K * sizeof(float), K, cudaMemcpyDeviceToDevice, stream) != cudaSuccess)
    return CONV2D_ECUDA;
  const int rc = launch();
  if (rc != CONV2D_OK) return rc;
  if (cudaEventRecord(ring.ev[slot], stream) != cudaSuccess) return CONV2D_ECUDA;
  return CONV2D_OK;
}

bool stream_capturing(cudaStream_t s) {
  cudaStreamCaptureStatus st = cudaStreamCaptureStatusNone;
  return cudaStreamIsCapturing(s, &st) == cudaSuccess && st != cudaStreamCaptureStatusNone;
}

template <int K, int U, int FSRC, int PF = 1, int GUARDS = 0>
int launch_single_v(const float *in, int H, int W, const float *filt, float *out, cudaStream_t stream, int band_h,
                    const DevInfo &dev, int min_band) {
  constexpr int CTAW = (FSRC == FSRC_CONST) ? 1 : kCtaWarps;
  auto kernel = k_conv2d_single<K, U, FSRC, CTAW, PF, GUARDS>;
  static std::atomic<int> occ_cache{0};
  SingleArgs a;
  a.in = in;
  a.filt = filt;
  a.out = out;
  a.H = H;
  a.W = W;
  a.Ho = H - K + 1;
  a.Wo = W - K + 1;
  a.n_cb = ceil_div(a.Wo, 128 * U);
  a.aligned = (aligned16(in) && (W % 4 == 0)) ? 1 : 0;
  if (band_h <= 0) {
    // one full wave of warp tiles: bands = resident warps / column blocks
    const long long resident_warps =
        static_cast<long long>(cta_occupancy(kernel, 0, occ_cache, CTAW)) * CTAW * dev.num_sms;
    const long long bands = resident_warps / a.n_cb > 0 ? resident_warps / a.n_cb : 1;
    band_h = ceil_div(a.Ho, bands);
    if (band_h < min_band) band_h = min_band;
  }
  if (band_h > a.Ho) band_h = a.Ho;
  a.band_h = band_h;
  const int n_bands = ceil_div(a.Ho, band_h);
  a.n_tiles = a.n_cb * n_bands;
  const int blocks = ceil_div(a.n_tiles, CTAW);
  auto go = [&]() {
    kernel<<<blocks, CTAW * kWarp, 0, stream>>>(a);
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  };
  if constexpr (FSRC == FSRC_CONST) return with_const_filter(filt, K, KCfg<K>::KP, stream, go);
  return go();
}

template <int K>
int launch_single(const float *in, int H, int W, const float *filt, float *out, cudaStream_t stream, int band_h,
                  const DevInfo &dev) {
  const int mb = g_min_band.load(std::memory_order_relaxed);
  const int min_band = mb > 0 ? mb : (K - 1 > 4 ? K - 1 : 4);
  const int v = g_variant.load(std::memory_order_relaxed);
  // CUDA-graph capture cannot use the event-guarded constant slots: shared-memory filter there
  const bool constant_ok = !stream_capturing(stream);
#define C2D_LS(UU, FS, PFF, G) launch_single_v<K, UU, FS, PFF, G>(in, H, W, filt, out, stream, band_h, dev, min_band)
  switch (v) {
    case 1: return C2D_LS(1, FSRC_SMEM, 1, 0);
    case 2: return C2D_LS(2, FSRC_SMEM, 1, 0);
    case 3: if (constant_ok) return C2D_LS(1, FSRC_CONST, 1, 0); break;
    case 4: if (constant_ok) return C2D_LS(2, FSRC_CONST, 1, 0); break;
    case 5: if (constant_ok) return C2D_LS(1, FSRC_CONST, 1, 1); break;
    case 6: if (constant_ok) return C2D_LS(1, FSRC_CONST, 1, 2); break;
    default: break;
  }
  // Tuned on B200 (tools/variants.py, profiles/): two 128-column
  // chunks per warp while K <= 7 (K = 9 on wide images); above, one chunk with a guarded prologue on
  // wide images (tall bands) and guarded prologue + epilogue on narrow ones (short bands, where the
  // wasted FMAs of an unguarded epilogue would be a large fraction).
  const bool u2 = (K <= 7) || (K <= 9 && W > 3000);
  if (!constant_ok) return u2 ? C2D_LS(2, FSRC_SMEM, 1, 0) : C2D_LS(1, FSRC_SMEM, 1, 0);
  if (u2) return C2D_LS(2, FSRC_CONST, 1, 0);
  if (W >= 4096) return C2D_LS(1, FSRC_CONST, 1, 1);
  return C2D_LS(1, FSRC_CONST, 1, 2);
#undef C2D_LS
}

// ------------------------------------------------------------------------------------------------
// multi channel
// ------------------------------------------------------------------------------------------------
template <int K>
struct MultiCfg {
  static constexpr int FB = (K <= 4) ? 8 : (K <= 8 ? 4 : 2);
};

template <int K, int FB>
int launch_multi_fb(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                    cudaStream_t stream, int band_h, const DevInfo &dev, size_t smem) {
  auto kernel = k_conv2d_multi<K, FB>;
  static std::atomic<int> occ_cache{0};
  static std::atomic<int> smem_set{0};
  if (smem > 48 * 1024 && smem_set.load() < static_cast<int>(smem)) {
    if (cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, dev.smem_optin) != cudaSuccess)
      return CONV2D_ECUDA;
    smem_set.store(dev.smem_optin);
  }
  MultiArgs a;
  a.in = in;
  a.filt = filt;
  a.out = out;
  a.N = N;
  a.C = C;
  a.H = H;
  a.W = W;
  a.F = F;
  a.Ho = H - K + 1;
  a.Wo = W - K + 1;
  a.n_cb = ceil_div(a.Wo, 128);
  a.n_fb = ceil_div(F, FB);
  a.aligned = (aligned16(in) && (W % 4 == 0)) ? 1 : 0;
  if (band_h <= 0) {
    // occupancy of this instantiation with this smem size (the cache holds the value for the
    // first smem size seen; good enough for choosing a band height)
    const long long resident_warps =
        static_cast<long long>(cta_occupancy(kernel, smem, occ_cache)) * kCtaWarps * dev.num_sms;
    const long long groups = static_cast<long long>(N) * a.n_fb * a.n_cb;
    long long bands = resident_warps / groups;
    if (bands < 1) bands = 1;
    band_h = ceil_div(a.Ho, bands);
    const int min_band = 4;
    if (band_h < min_band) band_h = min_band;
  }
  if (band_h > a.Ho) band_h = a.Ho;
  a.band_h = band_h;
  int n_bands = ceil_div(a.Ho, band_h);
  // all 4 warps of a CTA must share (n, F-block): pad the tiles per (n, F-block) to a multiple of 4
  while ((static_cast<long long>(a.n_cb) * n_bands) % kCtaWarps) ++n_bands;
  a.n_bands = n_bands;
  a.n_tiles = static_cast<long long>(N) * a.n_fb * n_bands * a.n_cb;
  const long long blocks = (a.n_tiles + kCtaWarps - 1) / kCtaWarps;
  if (blocks > 0x7fffffffLL) return CONV2D_ESHAPE;
  kernel<<<static_cast<unsigned>(blocks), kCtaWarps * kWarp, smem, stream>>>(a);
  return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
}

template <int K>
int launch_multi(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                 cudaStream_t stream, int band_h, const DevInfo &dev) {
  constexpr int FB = MultiCfg<K>::FB;
  constexpr int KP = KCfg<K>::KP;
  const size_t smem = static_cast<size_t>(C) * K * FB * KP * sizeof(float);
  if (smem <= static_cast<size_t>(dev.smem_optin))
    return launch_multi_fb<K, FB>(in, N, C, H, W, filt, F, out, stream, band_h, dev, smem);
  const size_t smem1 = static_cast<size_t>(C) * K * KP * sizeof(float);
  if (smem1 <= static_cast<size_t>(dev.smem_optin))
    return launch_multi_fb<K, 1>(in, N, C, H, W, filt, F, out, stream, band_h, dev, smem1);
  return CONV2D_ESHAPE;
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

}  // namespace

extern "C" {

int conv2d_single_ex(const float *in, int H, int W, const float *filt, int K, float *out, void *stream,
                     int band_h) {
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (int e = check_k(K)) return e;
  if (H < K || W < K) return CONV2D_ESHAPE;
  if (!aligned4(in) || !aligned4(filt) || !aligned4(out)) return CONV2D_EALIGN;
  const size_t in_b = static_cast<size_t>(H) * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(H - K + 1) * (W - K + 1) * sizeof(float);
  const size_t f_b = static_cast<size_t>(K) * K * sizeof(float);
  if (overlap(in, in_b, out, out_b) || overlap(filt, f_b, out, out_b)) return CONV2D_EOVERLAP;
  DevInfo dev;
  if (current_device_info(&dev)) return CONV2D_ECUDA;
  cudaStream_t s = static_cast<cudaStream_t>(stream);
#define C2D_CALL_SINGLE(KK) launch_single<KK>(in, H, W, filt, out, s, band_h, dev)
  C2D_K_SWITCH(K, C2D_CALL_SINGLE)
#undef C2D_CALL_SINGLE
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
#define C2D_CALL_MULTI(KK) launch_multi<KK>(in, N, C, H, W, filt, F, out, s, band_h, dev)
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
    default: return "unknown error code";
  }
}

int conv2d_version(void) { return 100; }

// Not part of include/conv2d.h: selects a kernel variant for tuning tools (0 = default).
int c2d_debug_set_variant(int v) {
  const int old = g_variant.exchange(v);
  return old;
}

// Not part of include/conv2d.h: minimum band height override for tuning tools (0 = default).
int c2d_debug_set_min_band(int v) {
  const int old = g_min_band.exchange(v);
  return old;
}

}  // extern "C"

// common.h -- declarations shared by the C-ABI unit (conv2d_capi.cu) and the per-K launch units
// (inst_kNN.cu): device info, tuning overrides, and the per-K launch entry points.
#pragma once

#include <atomic>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"

namespace c2d {

constexpr int kMaxDevices = 64;

struct DevInfo {
  int id = 0;  // CUDA device ordinal (the current device of the call)
  int num_sms = 0;
  int smem_optin = 0;
};

// Tuning overrides exist only in the tuning build (-DC2D_TUNING, libconv2d_tune.so: every kernel
// variant instantiated, selectable through c2d_debug_set_*); the product libconv2d.so has the tuned
// defaults only and no process-global switches.
#ifdef C2D_TUNING
extern std::atomic<int> g_variant;    // single-channel kernel variant (0 = tuned default)
extern std::atomic<int> g_min_band;   // minimum band height of the automatic band choice
extern std::atomic<int> g_mvariant;   // multi-channel kernel variant
inline int tuning_variant() { return g_variant.load(std::memory_order_relaxed); }
inline int tuning_min_band() { return g_min_band.load(std::memory_order_relaxed); }
inline int tuning_mvariant() { return g_mvariant.load(std::memory_order_relaxed); }
#else
constexpr int tuning_variant() { return 0; }
constexpr int tuning_min_band() { return 0; }
constexpr int tuning_mvariant() { return 0; }
#endif

// Stream-ordered scratch memory from a library-owned memory pool of the current device (release
// threshold "never", so the pool keeps its memory across synchronisations instead of returning it to
// the driver -- the default pool trims at every sync, which turns each call into a real allocation).
// Release with cudaFreeAsync on a stream ordered after the last use.
cudaError_t scratch_alloc(void **p, size_t bytes, cudaStream_t stream);
cudaError_t scratch_trim();

// band_h value for single_entry: automatic band height, and never the filter-row split kernel (its
// sums are grouped differently; conv2d_single_pad's border strips must match the one-tile kernel bits)
constexpr int kBandNoSplit = -2;
// ... and with the per-CTA shared-memory filter (no constant-slot staging: a call on a side stream
// must not wait for the slot's previous user on the main stream)
constexpr int kBandSmemFilter = -3;

// per-K entry points, explicitly instantiated one K per translation unit (csrc/inst_kNN.cu)
// N images of H x W (input image stride H*P floats, output image stride (H-K+1)*Po floats); rows
// >= H1 at in2 (H1 == H: one segment; N == 1 when H1 < H); input / output row pitch P / Po floats
template <int K>
int single_entry(const float *in, int N, int H, int W, const float *filt, float *out, cudaStream_t stream,
                 int band_h, const DevInfo &dev, const float *in2, int H1, long long P, int Po);
// Rectangular KH x KW filters (KH a template parameter: one translation unit per KH, inst_rect_khNN.cu)
template <int KH>
int rect_entry(const float *in, int H, int W, const float *filt, int KW, float *out, cudaStream_t stream,
               const DevInfo &dev);
template <int K>
int multi_entry(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                cudaStream_t stream, int band_h, const DevInfo &dev);

}  // namespace c2d

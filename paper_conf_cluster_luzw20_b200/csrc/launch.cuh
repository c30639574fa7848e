// launch.cuh -- host-side launch code of the kernels for one K (included once per translation unit
// csrc/inst_kNN.cu): launch geometry (band height, F-block, segments), filter staging (constant slot
// or shared memory), kernel-variant selection. State (constant-slot events, occupancy caches) has
// internal linkage: one copy per unit, i.e. per K, matching the per-unit constant banks.
#pragma once

#include <atomic>
#include <cstdint>
#include <mutex>

#include <cuda_runtime.h>

#include "common.h"
#include "conv2d_kernels.cuh"
#include "conv2d_multi.cuh"
#include "conv2d_split.cuh"
#include "conv2d_wide.cuh"
#include "conv2d_pair.cuh"
#include "conv2d_mob.cuh"

namespace {

using namespace c2d;

bool aligned16(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 15u) == 0; }

int ceil_div(long long a, long long b) { return static_cast<int>((a + b - 1) / b); }

// Occupancy (CTAs per SM) of one kernel instantiation, cached per dynamic shared-memory size (the
// devices of one box are identical B200s; the smem size depends on call arguments such as C). A few
// lock-free entries (smem << 16 | value); a miss past the last entry just recomputes.
struct OccCache {
  std::atomic<long long> e[8] = {};
};
template <typename KernelT>
int cta_occupancy(KernelT kernel, size_t dyn_smem, OccCache &cache, int cta_threads) {
  const long long key = static_cast<long long>(dyn_smem) << 16;
  for (auto &slot : cache.e) {
    const long long v = slot.load(std::memory_order_relaxed);
    if (v == 0) break;
    if ((v & ~0xffffLL) == key) return static_cast<int>(v & 0xffff);
  }
  int blocks = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, kernel, cta_threads, dyn_smem) != cudaSuccess ||
      blocks < 1)
    blocks = 1;
  for (auto &slot : cache.e) {
    long long expect = 0;
    if (slot.compare_exchange_strong(expect, key | blocks, std::memory_order_relaxed)) break;
    if ((expect & ~0xffffLL) == key) break;
  }
  return blocks;
}

// Opt a kernel instantiation into more than 48 KiB of dynamic shared memory, once per DEVICE (the
// attribute is per device; a process may drive several GPUs).
struct SmemOptIn {
  std::atomic<int> done[kMaxDevices] = {};
};
template <typename KernelT>
int ensure_smem(KernelT kernel, size_t smem, const DevInfo &dev, SmemOptIn &flag) {
  if (smem <= 48 * 1024) return CONV2D_OK;
  if (smem > static_cast<size_t>(dev.smem_optin)) return CONV2D_ESHAPE;
  if (dev.id < 0 || dev.id >= kMaxDevices) return CONV2D_ECUDA;
  if (flag.done[dev.id].load(std::memory_order_acquire)) return CONV2D_OK;
  if (cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, dev.smem_optin) != cudaSuccess)
    return CONV2D_ECUDA;
  flag.done[dev.id].store(1, std::memory_order_release);
  return CONV2D_OK;
}

// Band count per image. band_h > 0 (explicit): ceil(Ho / band_h) bands. Automatic: a wave-quantisation
// cost model over the n_img x n_cb x bands tiles with `resident` tiles per wave: a tile of h output
// rows streams h + K - 1 input rows (Alg. 2 case 1 is K-1 rows of prologue), and the grid runs in
// ceil(tiles / resident) waves, so pick the band count b minimising waves(b) * (ceil(Ho / b) + K - 1)
// with bands at least min_band rows tall. (One image: one full wave of bands, the round-1 choice; a
// batch of large images: several waves of taller bands instead of an under-filled single wave --
// 8 x 8192^2 K=15: 4 bands per image filled 86% of one wave.) Bands are balanced (band_start).
int band_count(int Ho, int K, int n_cb, int n_img, long long resident, int band_h, int min_band) {
  if (band_h > 0) {
    long long b = (Ho + static_cast<long long>(band_h) - 1) / band_h;
    return static_cast<int>(b < 1 ? 1 : (b > Ho ? Ho : b));
  }
  const long long groups = static_cast<long long>(n_cb) * n_img;
  long long bmax = min_band > 1 ? Ho / min_band : Ho;
  if (bmax < 1) bmax = 1;
  if (bmax > 8192) bmax = 8192;
  if (resident < 1) resident = 1;
  long long best_b = 1;
  double best = 1e300;
  for (long long b = 1; b <= bmax; ++b) {
    const long long h = (Ho + b - 1) / b;
    const long long waves = (groups * b + resident - 1) / resident;
    const double cost = static_cast<double>(waves) * static_cast<double>(h + K - 1);
    if (cost < best * (1.0 - 1e-9)) {  // ties: the fewest bands
      best = cost;
      best_b = b;
    }
  }
  return static_cast<int>(best_b);
}

// ------------------------------------------------------------------------------------------------
// single channel
// ------------------------------------------------------------------------------------------------
// Tuning build only (c2d_debug_set_variant; 0 = the tuned default):
//   1: filter in shared memory, U=1 (4 warps/CTA)     2: shared memory, U=2
//   3: filter in a __constant__ slot, U=1 (1 warp/CTA) 4: __constant__ slot, U=2
//   5-9, 13, 15: guard / prefetch variants of the constant-slot kernel (see launch_single)
//   10-12: filter-row split over G parts (conv2d_split.cuh)

// Constant-bank filter slot of this unit (this K), per device: it holds the filter of the last call
// with this K. A call waits (stream-ordered) for the event recorded behind the previous kernel that
// read the slot before overwriting it, so calls on different streams never see each other's filter;
// calls with the same K on different streams are serialised by that wait, calls on one stream cost
// nothing.
struct ConstRing {
  std::mutex mu;
  bool init = false;
  float *base = nullptr;  // device address of c_filt
  cudaEvent_t ev;
};
ConstRing g_cring[kMaxDevices];

template <typename LaunchFn>
int with_const_filter(const float *filt, int K, int KP, cudaStream_t stream, const DevInfo &dev, LaunchFn launch) {
  if (dev.id < 0 || dev.id >= kMaxDevices) return CONV2D_ECUDA;
  ConstRing &ring = g_cring[dev.id];
  std::lock_guard<std::mutex> lk(ring.mu);
  if (!ring.init) {
    void *p = nullptr;
    if (cudaGetSymbolAddress(&p, c_filt) != cudaSuccess) return CONV2D_ECUDA;
    ring.base = static_cast<float *>(p);
    if (cudaEventCreateWithFlags(&ring.ev, cudaEventDisableTiming) != cudaSuccess) return CONV2D_ECUDA;
    ring.init = true;
  }
  if (cudaStreamWaitEvent(stream, ring.ev, 0) != cudaSuccess) return CONV2D_ECUDA;
  // K rows of K floats -> K rows of KP floats (16-byte aligned rows for LDCU.128)
  if (cudaMemcpy2DAsync(ring.base, KP * sizeof(float), filt, K * sizeof(float), K * sizeof(float), K,
                        cudaMemcpyDeviceToDevice, stream) != cudaSuccess)
    return CONV2D_ECUDA;
  const int rc = launch();
  if (rc != CONV2D_OK) return rc;
  if (cudaEventRecord(ring.ev, stream) != cudaSuccess) return CONV2D_ECUDA;
  return CONV2D_OK;
}

bool stream_capturing(cudaStream_t s) {
  cudaStreamCaptureStatus st = cudaStreamCaptureStatusNone;
  return cudaStreamIsCapturing(s, &st) == cudaSuccess && st != cudaStreamCaptureStatusNone;
}

// Geometry shared by the one-warp-tile and the split launches.
struct SingleGeom {
  const float *in, *in2;
  int N, H, W, H1;
  long long P;
  int Po;
};

template <typename ArgsT>
void fill_args(ArgsT &a, const SingleGeom &g, int K, int U, float *out) {
  a.in = g.in;
  a.in2 = g.in2;
  a.H1 = g.H1;
  a.P = static_cast<int>(g.P);
  a.Wc = static_cast<int>(g.P);
  a.Po = g.Po;
  a.out = out;
  a.H = g.H;
  a.W = g.W;
  a.Ho = g.H - K + 1;
  a.Wo = g.W - K + 1;
  a.n_img = g.N;
  a.img_in = static_cast<long long>(g.H) * g.P;
  a.img_out = static_cast<long long>(a.Ho) * g.Po;
  a.n_cb = ceil_div(a.Wo, 128 * U);
  a.aligned = (aligned16(g.in) && aligned16(g.in2) && (g.P % 4 == 0)) ? 1 : 0;
}

template <int K, int U, int FSRC, int PF = 1, int GUARDS = 0, bool HALO = false>
int launch_single_v(const SingleGeom &g, const float *filt, float *out, cudaStream_t stream, int band_h,
                    const DevInfo &dev, int min_band) {
  constexpr int CTAW = (FSRC == FSRC_CONST) ? 1 : kCtaWarps;
  auto kernel = k_conv2d_single<K, U, FSRC, CTAW, PF, GUARDS, HALO>;
  static OccCache occ_cache;
  const size_t ring = (PF >= 3) ? CTAW * RowRing<K, U, kWarp, (PF >= 3 ? PF : 2)>::kBytes : 0;
  SingleArgs a;
  fill_args(a, g, K, U, out);
  a.filt = filt;
  const long long resident = static_cast<long long>(cta_occupancy(kernel, ring, occ_cache, CTAW * kWarp)) * CTAW *
                             dev.num_sms;
  a.n_bands = band_count(a.Ho, K, a.n_cb, a.n_img, resident, band_h, min_band);
  const long long tiles = static_cast<long long>(a.n_cb) * a.n_bands * a.n_img;
  if (tiles > 0x7fffffffLL - CTAW) return CONV2D_ESHAPE;
  a.n_tiles = static_cast<int>(tiles);
  const int blocks = ceil_div(a.n_tiles, CTAW);
  auto go = [&]() {
    kernel<<<blocks, CTAW * kWarp, ring, stream>>>(a);
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  };
  if constexpr (FSRC == FSRC_CONST) return with_const_filter(filt, K, KCfg<K>::KP, stream, dev, go);
  return go();
}

// Wide-lane kernel (conv2d_wide.cuh): 8 contiguous columns per lane, 256-column warp tiles, one warp
// per CTA.
template <int K, int FSRC, int PF, int GUARDS, bool HALO = false>
int launch_wide_v(const SingleGeom &g, const float *filt, float *out, cudaStream_t stream, int band_h,
                  const DevInfo &dev, int min_band) {
  auto kernel = k_conv2d_wide<K, K, FSRC, PF, GUARDS, HALO>;
  static OccCache occ_cache;
  const size_t ring = (PF >= 3) ? WideRing<K, (PF >= 3 ? PF : 2)>::kBytes : 0;
  SingleArgs a;
  fill_args(a, g, K, 2, out);  // n_cb in 256-column blocks (= two 128-column chunks)
  a.filt = filt;
  const long long resident = static_cast<long long>(cta_occupancy(kernel, ring, occ_cache, kWarp)) * dev.num_sms;
  a.n_bands = band_count(a.Ho, K, a.n_cb, a.n_img, resident, band_h, min_band);
  const long long tiles = static_cast<long long>(a.n_cb) * a.n_bands * a.n_img;
  if (tiles > 0x7fffffffLL) return CONV2D_ESHAPE;
  a.n_tiles = static_cast<int>(tiles);
  auto go = [&]() {
    kernel<<<a.n_tiles, kWarp, ring, stream>>>(a);
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  };
  if constexpr (FSRC == FSRC_CONST) return with_const_filter(filt, K, KCfg<K>::KP, stream, dev, go);
  return go();
}

// Slot-paired FFMA2 kernel (conv2d_pair.cuh), odd K: the constant slot holds the pair table
//   pairs [p][j] = (f[H+p][j], f[p][j]), single [j] = f[H-1][j]
// built by three stream-ordered copies (two interleave 4-byte elements at an 8-byte destination pitch),
// recycled with the slot's event like the plain filter staging.
template <int K, typename LaunchFn>
int with_const_pair_filter(const float *filt, cudaStream_t stream, const DevInfo &dev, LaunchFn launch) {
  using PC = PairCfg<K>;
  if (dev.id < 0 || dev.id >= kMaxDevices) return CONV2D_ECUDA;
  ConstRing &ring = g_cring[dev.id];
  std::lock_guard<std::mutex> lk(ring.mu);
  if (!ring.init) {
    void *p = nullptr;
    if (cudaGetSymbolAddress(&p, c_filt) != cudaSuccess) return CONV2D_ECUDA;
    ring.base = static_cast<float *>(p);
    if (cudaEventCreateWithFlags(&ring.ev, cudaEventDisableTiming) != cudaSuccess) return CONV2D_ECUDA;
    ring.init = true;
  }
  if (cudaStreamWaitEvent(stream, ring.ev, 0) != cudaSuccess) return CONV2D_ECUDA;
  const size_t n = static_cast<size_t>(PC::NP) * K;
  if (cudaMemcpy2DAsync(ring.base, 8, filt + PC::H * K, 4, 4, n, cudaMemcpyDeviceToDevice, stream) != cudaSuccess ||
      cudaMemcpy2DAsync(ring.base + 1, 8, filt, 4, 4, n, cudaMemcpyDeviceToDevice, stream) != cudaSuccess ||
      cudaMemcpyAsync(ring.base + PC::kSingle, filt + (PC::H - 1) * K, K * sizeof(float), cudaMemcpyDeviceToDevice,
                      stream) != cudaSuccess)
    return CONV2D_ECUDA;
  const int rc = launch();
  if (rc != CONV2D_OK) return rc;
  if (cudaEventRecord(ring.ev, stream) != cudaSuccess) return CONV2D_ECUDA;
  return CONV2D_OK;
}

template <int K, int PF, bool HALO = false>
int launch_pair_v(const SingleGeom &g, const float *filt, float *out, cudaStream_t stream, int band_h,
                  const DevInfo &dev, int min_band) {
  auto kernel = k_conv2d_pair<K, PF, HALO>;
  static OccCache occ_cache;
  const size_t ring = (PF >= 3) ? RowRing<K, 1, kWarp, (PF >= 3 ? PF : 2)>::kBytes : 0;
  SingleArgs a;
  fill_args(a, g, K, 1, out);
  a.filt = filt;
  const long long resident = static_cast<long long>(cta_occupancy(kernel, ring, occ_cache, kWarp)) * dev.num_sms;
  a.n_bands = band_count(a.Ho, K, a.n_cb, a.n_img, resident, band_h, min_band);
  const long long tiles = static_cast<long long>(a.n_cb) * a.n_bands * a.n_img;
  if (tiles > 0x7fffffffLL) return CONV2D_ESHAPE;
  a.n_tiles = static_cast<int>(tiles);
  return with_const_pair_filter<K>(filt, stream, dev, [&]() {
    kernel<<<a.n_tiles, kWarp, ring, stream>>>(a);
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  });
}

// Rectangular KH x KW filters (conv2d_single_rect): the wide-lane kernel with a KH-slot
// ring and a KW-wide window, filter staged per CTA in shared memory, one row in flight in registers.
template <int KH, int KW>
int launch_rect_v(const float *in, int H, int W, const float *filt, float *out, cudaStream_t stream,
                  const DevInfo &dev) {
  auto kernel = k_conv2d_wide<KH, KW, FSRC_SMEM, 1, 0, false>;
  static OccCache occ_cache;
  SingleArgs a;
  const SingleGeom g{in, in, 1, H, W, H, W, W - KW + 1};
  fill_args(a, g, KH, 2, out);  // Ho from KH
  a.Wo = W - KW + 1;
  a.img_out = static_cast<long long>(a.Ho) * a.Po;
  a.n_cb = ceil_div(a.Wo, kWideSpan);
  a.filt = filt;
  const long long resident = static_cast<long long>(cta_occupancy(kernel, 0, occ_cache, kWarp)) * dev.num_sms;
  const bool tiny = static_cast<long long>(H) * W <= 512LL * 512;
  const int min_band = tiny ? 1 : (KH - 1 > 4 ? KH - 1 : 4);
  a.n_bands = band_count(a.Ho, KH, a.n_cb, 1, resident, 0, min_band);
  const long long tiles = static_cast<long long>(a.n_cb) * a.n_bands;
  if (tiles > 0x7fffffffLL) return CONV2D_ESHAPE;
  a.n_tiles = static_cast<int>(tiles);
  kernel<<<a.n_tiles, kWarp, 0, stream>>>(a);
  return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
}

// Filter-row split (conv2d_split.cuh): same tile geometry as launch_single_v, but a tile takes G
// warps -- a cluster of G one-warp CTAs (CL = 1) or one CTA of G warps (CL = 0) -- so a full wave has
// G times fewer, taller bands.
template <int K, int G, int U, int PF, int R, int GUARDS, int CL>
int launch_split_v(const SingleGeom &g, const float *filt, float *out, cudaStream_t stream, int band_h,
                   const DevInfo &dev, int min_band) {
  static_assert(G >= 1 && G <= 8 && G <= K, "portable cluster of at most K CTAs");
  auto kernel = k_conv2d_split<K, G, U, PF, R, GUARDS, CL>;
  static OccCache occ_cache;  // CL = 1: resident clusters per GPU; CL = 0: CTAs per SM
  static SmemOptIn smem_flag;
  const size_t smem = static_cast<size_t>(SplitSmem<K, U, PF, R>::kPart) * (CL ? 1 : G);
  const int threads = CL ? kWarp : G * kWarp;
  SplitArgs a;
  fill_args(a, g, K, U, out);
  if (int e = ensure_smem(kernel, smem, dev, smem_flag)) return e;
  cudaLaunchConfig_t cfg = {};
  cfg.blockDim = dim3(threads, 1, 1);
  cfg.dynamicSmemBytes = smem;
  cfg.stream = stream;
  cudaLaunchAttribute attr[1];
  attr[0].id = cudaLaunchAttributeClusterDimension;
  attr[0].val.clusterDim.x = G;
  attr[0].val.clusterDim.y = 1;
  attr[0].val.clusterDim.z = 1;
  cfg.attrs = attr;
  cfg.numAttrs = CL ? 1 : 0;
  long long resident = 1;
  if (band_h <= 0) {
    // resident tiles of one full wave (clusters: as the cluster scheduler places them)
    int v = 0;
    const long long key = static_cast<long long>(smem) << 16;
    const long long cached = occ_cache.e[0].load(std::memory_order_relaxed);
    if (cached != 0 && (cached & ~0xffffLL) == key) {
      v = static_cast<int>(cached & 0xffff);
    } else {
      if constexpr (CL) {
        cfg.gridDim = dim3(G * dev.num_sms, 1, 1);
        int clusters = 0;
        if (cudaOccupancyMaxActiveClusters(&clusters, kernel, &cfg) != cudaSuccess || clusters < 1) clusters = 1;
        v = clusters;
      } else {
        int blocks = 0;
        if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, kernel, threads, smem) != cudaSuccess ||
            blocks < 1)
          blocks = 1;
        v = blocks * dev.num_sms;
      }
      occ_cache.e[0].store(key | v, std::memory_order_relaxed);
    }
    resident = v;
  }
  a.n_bands = band_count(a.Ho, K, a.n_cb, a.n_img, resident, band_h, min_band);
  const long long tiles = static_cast<long long>(a.n_cb) * a.n_bands * a.n_img;
  if (tiles * G > 0x7fffffffLL) return CONV2D_ESHAPE;
  a.n_tiles = static_cast<int>(tiles);
  cfg.gridDim = dim3(static_cast<unsigned>(CL ? tiles * G : tiles), 1, 1);
  auto go = [&]() {
    if (cudaLaunchKernelEx(&cfg, kernel, a) != cudaSuccess) {
      (void)cudaGetLastError();  // launch-configuration errors are not sticky: do not leak into the next call
      return CONV2D_ECUDA;
    }
    return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
  };
  return with_const_filter(filt, K, KCfg<K>::KP, stream, dev, go);
}

// The tuned default kernel choice (HALO: conv2d_single_halo's two-segment row addressing, same choice
// and so the same bits as the one-segment call on the concatenated rows).
template <int K, bool HALO>
int launch_single_default(const SingleGeom &g, const float *filt, float *out, cudaStream_t stream, int band_h,
                          const DevInfo &dev, int min_band, bool constant_ok) {
#define C2D_LS(UU, FS, PFF, G) launch_single_v<K, UU, FS, PFF, G, HALO>(g, filt, out, stream, band_h, dev, min_band)
#define C2D_LW(FS, PFF, G) launch_wide_v<K, FS, PFF, G, HALO>(g, filt, out, stream, band_h, dev, min_band)
#define C2D_SP(GG, UU, PFF, RR, CLL) launch_split_v<K, GG, UU, PFF, RR, 1, CLL>(g, filt, out, stream, band_h, dev, 1)
  const int W = g.W;
  const bool force_smem = band_h == kBandSmemFilter;
  const bool no_split = band_h == kBandNoSplit || force_smem;  // internal callers: the one-tile kernel's bits
  if (no_split) band_h = 0;
  // Narrow images with large K (latency regime: a full wave of one-warp tiles leaves bands of a few
  // rows, and the K-1 prologue rows of Alg. 2 case 1 dominate): filter rows split over a cluster of 2
  // one-warp CTAs (tools/split_sweep.py: 1024^2 K=15 24 -> 30 Gpx/s, 256^2 K=15 1.6 -> 3.8).
  // Keyed on (W, K) only, so row bands of one image (same W) take the same kernel: bitwise seams.
  if constexpr (K >= 11) {
    if (constant_ok && W <= 1024 && !no_split) return C2D_SP(2, 1, 4, 4, 1);
  }
#undef C2D_SP
  // Tuned on B200 (tools/variants.py sweeps, profiles/r02e_variants*.txt):
  //   K <= 3        the wide-lane kernel (8 contiguous columns per lane): constant-slot filter on wide
  //                 images, per-CTA shared-memory filter below (no slot staging: 4096^2 511 vs 444 Gpx/s);
  //   K = 4, 5      images up to 2048 wide: wide lanes + shared-memory filter; wider: two 128-column
  //                 chunks per warp with a 4-stage cp.async row ring;
  //   K = 6..9      W >= 8192: wide lanes, both Alg. 2 edge cases guarded (8192^2 K=9 325 vs 307 Gpx/s,
  //                 K=7 457 vs 449; batches of 8: 340 vs 335, 503 vs 491); narrower: one or two chunks +
  //                 ring + guards;
  //   K = 10, 11    one chunk + ring + guards;
  //   K >= 12       one chunk (the wide kernel's 32 KB loop body overflows the instruction cache at
  //                 K >= 11: ncu no_instructions 20% at K=15), register row fetch, guarded prologue on
  //                 wide images, guarded prologue + epilogue on narrow ones.
  // Small images with K < 11 are latency-bound (a few microseconds): the per-CTA shared-memory filter
  // skips the constant-slot staging (a stream-ordered copy plus two event operations, ~3 us of host
  // and device time per call, tools/host_overhead.py). Same summation order, same bits.
  const long long px = static_cast<long long>(g.H) * W * g.N;  // input pixels of the launch (all images)
  const bool small = px <= 512LL * 512 || (K <= 5 && px <= 1024LL * 1024);
  // Launches with >= 32 M (128 M) input pixels amortise the constant-slot staging (a stream-ordered copy
  // + event ops, ~3 us) and take the constant-filter kernels that win on long launches; shorter ones
  // keep the per-CTA shared-memory filter (profiles/r02q_all_b8.txt: batches of 8; r02c/r02e/r02l: one
  // image).
  const bool big = px >= (32LL << 20), giant = px >= (128LL << 20);
  const bool cst = constant_ok && !force_smem;
  if constexpr (K <= 3) {
    // wide lanes; constant slot on long launches (4096^2 x8 686 vs 642 Gpx/s), shared memory otherwise
    // (one 4096^2 image 511 vs 442)
    if (cst && W >= 4096 && big) return C2D_LW(FSRC_CONST, 1, 0);
    return C2D_LW(FSRC_SMEM, 1, 0);
  }
  if constexpr (K <= 5) {
    // two chunks (FFMA2) + ring + guards on launches >= 16 M pixels (x8: 8192^2 711 vs 649, 2048^2 536 vs
    // 466; one 4096^2 image 467 vs 419), wide lanes + shared memory below (one 2048^2 image 227 vs 217)
    if (cst && px >= (16LL << 20) && W >= 2048) return C2D_LS(2, FSRC_CONST, 4, 2);
    if (!cst || W <= 2048) return C2D_LW(FSRC_SMEM, 1, 0);
  }
  if (!cst || (K < 11 && small)) {
    if constexpr (K <= 7) return C2D_LS(2, FSRC_SMEM, 1, 0);
    else return C2D_LS(1, FSRC_SMEM, 1, 0);
  }
  if constexpr (K <= 5) {
    return C2D_LS(2, FSRC_CONST, 4, 0);
  } else if constexpr (K <= 7) {
    // slot-paired FFMA2 ring on the longest launches (r02r: 8 x 8192^2 K=7 528 vs 511 Gpx/s)
    if constexpr (K == 7) {
      if (W >= 8192 && giant) return launch_pair_v<K, 4, HALO>(g, filt, out, stream, band_h, dev, min_band);
    }
    if (W >= 8192) return C2D_LW(FSRC_CONST, 1, 2);
    if (big) return C2D_LW(FSRC_CONST, 1, 0);  // x8: 4096^2 486 vs 449, 2048^2 402 vs 374
    if (W >= 4096) return C2D_LS(2, FSRC_CONST, 4, 2);
    return C2D_LS(1, FSRC_CONST, 4, 2);
  } else if constexpr (K <= 9) {
    if (W >= 8192 && giant) return C2D_LS(2, FSRC_CONST, 1, 0);  // x8 349 vs 338 (one image: -11%)
    if (W >= 8192) return C2D_LW(FSRC_CONST, 1, 2);
    return C2D_LS(1, FSRC_CONST, 4, 2);
  } else if constexpr (K <= 11) {
    // two chunks with FFMA2 (row_step1) on images >= 4096 wide (profiles/r02l_ffma2*.txt: 8192^2 K=11
    // x8 246 vs 231 Gpx/s)
    if (W >= 4096) return C2D_LS(2, FSRC_CONST, 1, 2);
    return C2D_LS(1, FSRC_CONST, 4, 2);
  } else {
    // K = 12-14, wide: the cp.async ring with the guarded prologue (variant 15: 8192^2 K=13 155 -> 161
    // Gpx/s, 4096^2 128 -> 132); K = 15 measured equal either way and keeps the register row fetch.
    // Two chunks with FFMA2 at 8192 (K <= 13: x8 178 vs 171); below 4096 two chunks for short launches,
    // the one-chunk ring on long ones (2048^2 K=15 x8 107 vs 101).
    // K = 15 on long launches >= 4096 wide: the slot-paired FFMA2 ring (conv2d_pair.cuh; r02r: 8 x 8192^2
    // 132 vs 124 Gpx/s, 8 x 4096^2 125 vs 118, one 8192^2 image 122 vs 117)
    if constexpr (K == 15) {
      if (W >= 4096 && big) return launch_pair_v<K, 4, HALO>(g, filt, out, stream, band_h, dev, min_band);
    }
    if (K <= 13 && W >= 8192) return C2D_LS(2, FSRC_CONST, 1, 2);
    if (K <= 14 && W >= 4096) return C2D_LS(1, FSRC_CONST, 4, 1);
    if (W >= 4096) return C2D_LS(1, FSRC_CONST, 1, 1);
    if (big) return C2D_LS(1, FSRC_CONST, 4, 1);
    return C2D_LS(2, FSRC_CONST, 1, 2);
  }
#undef C2D_LS
#undef C2D_LW
}

template <int K>
int launch_single(const SingleGeom &g, const float *filt, float *out, cudaStream_t stream, int band_h,
                  const DevInfo &dev) {
  const int mb = tuning_min_band();
  // Minimum band height K-1 (>= 4) bounds the Alg. 2 case-1 overhead once a wave is full; images up
  // to 512^2 cannot fill a wave even with one-row bands, and there the latency of a band's row chain
  // dominates: no minimum (tools/latency.py, one 256^2 call: K=3 10.3 -> 8.9 us, K=9 20.7 -> 14.2 us,
  // K=15 smem path 42 -> 28.6 us). Band height never changes the bits.
  const bool tiny = static_cast<long long>(g.H) * g.W * g.N <= 512LL * 512;
  const int min_band = mb > 0 ? mb : (tiny ? 1 : (K - 1 > 4 ? K - 1 : 4));
  // CUDA-graph capture cannot use the event-guarded constant slots: shared-memory filter there
  const bool constant_ok = !stream_capturing(stream);
  if (g.H1 < g.H) return launch_single_default<K, true>(g, filt, out, stream, band_h, dev, min_band, constant_ok);
#ifdef C2D_TUNING
#define C2D_LS(UU, FS, PFF, G) launch_single_v<K, UU, FS, PFF, G>(g, filt, out, stream, band_h, dev, min_band)
  switch (tuning_variant()) {
    case 1: return C2D_LS(1, FSRC_SMEM, 1, 0);
    case 2: return C2D_LS(2, FSRC_SMEM, 1, 0);
    case 3: if (constant_ok) return C2D_LS(1, FSRC_CONST, 1, 0); break;
    case 4: if (constant_ok) return C2D_LS(2, FSRC_CONST, 1, 0); break;
    case 5: if (constant_ok) return C2D_LS(1, FSRC_CONST, 1, 1); break;
    case 6: if (constant_ok) return C2D_LS(1, FSRC_CONST, 1, 2); break;
    case 7: if (constant_ok) return C2D_LS(2, FSRC_CONST, 4, 0); break;
    case 8: if (constant_ok) return C2D_LS(2, FSRC_CONST, 8, 0); break;
    case 9: if (constant_ok) return C2D_LS(1, FSRC_CONST, 4, 2); break;
    case 13: if constexpr (K >= 5 && K <= 9) { if (constant_ok) return C2D_LS(2, FSRC_CONST, 4, 2); } break;
    case 15: if constexpr (K >= 10) { if (constant_ok) return C2D_LS(1, FSRC_CONST, 4, 1); } break;
    case 16: if (constant_ok) return C2D_LS(1, FSRC_CONST, 2, 1); break;
    case 17: if (constant_ok) return C2D_LS(1, FSRC_CONST, 2, 0); break;
    case 18: if (constant_ok) return C2D_LS(2, FSRC_CONST, 2, 0); break;
    case 19: if (constant_ok) return C2D_LS(1, FSRC_CONST, 2, 2); break;
    case 40: if (constant_ok) return C2D_LS(2, FSRC_CONST, 1, 1); break;
    case 41: if (constant_ok) return C2D_LS(2, FSRC_CONST, 4, 1); break;
    case 42: if (constant_ok) return C2D_LS(2, FSRC_CONST, 1, 2); break;
    case 43: if (constant_ok) return C2D_LS(2, FSRC_CONST, 4, 2); break;
    // slot-paired FFMA2 ring (conv2d_pair.cuh), odd K
    case 48: if constexpr (K % 2 == 1 && K >= 3) { if (constant_ok) return launch_pair_v<K, 1>(g, filt, out, stream, band_h, dev, min_band); } break;
    case 49: if constexpr (K % 2 == 1 && K >= 3) { if (constant_ok) return launch_pair_v<K, 4>(g, filt, out, stream, band_h, dev, min_band); } break;
    default: break;
  }
#undef C2D_LS
  // wide-lane kernel (conv2d_wide.cuh; variants 20-26)
#define C2D_LW(FS, PFF, G) launch_wide_v<K, FS, PFF, G>(g, filt, out, stream, band_h, dev, min_band)
  switch (tuning_variant()) {
    case 20: if (constant_ok) return C2D_LW(FSRC_CONST, 1, 0); break;
    case 21: if (constant_ok) return C2D_LW(FSRC_CONST, 1, 1); break;
    case 22: if (constant_ok) return C2D_LW(FSRC_CONST, 1, 2); break;
    case 23: if (constant_ok) return C2D_LW(FSRC_CONST, 4, 0); break;
    case 24: if (constant_ok) return C2D_LW(FSRC_CONST, 4, 1); break;
    case 25: if (constant_ok) return C2D_LW(FSRC_CONST, 4, 2); break;
    case 26: return C2D_LW(FSRC_SMEM, 1, 0);
    case 27: if (constant_ok) return C2D_LW(FSRC_CONST, 2, 0); break;
    case 28: if (constant_ok) return C2D_LW(FSRC_CONST, 2, 2); break;
    case 29: return C2D_LW(FSRC_SMEM, 2, 0);
    default: break;
  }
#undef C2D_LW
  // filter-row split (conv2d_split.cuh; variants 10-12)
#define C2D_SP(GG, UU, PFF, RR, CLL) launch_split_v<K, GG, UU, PFF, RR, 1, CLL>(g, filt, out, stream, band_h, dev, 1)
  const int v = tuning_variant();
  if (constant_ok && v >= 10 && v <= 12) {
    if constexpr (K >= 3) {
      switch (v) {
        case 10: return C2D_SP(2, 1, 4, 4, 1);  // cluster of 2 one-warp CTAs (the default below)
        case 11: return C2D_SP(2, 1, 4, 8, 0);  // one CTA of 2 warps (same sums: same bits as 10)
        case 12: return C2D_SP(3, 1, 4, 8, 0);  // one CTA of 3 warps
        default: break;
      }
    }
  }
#undef C2D_SP
#endif
  return launch_single_default<K, false>(g, filt, out, stream, band_h, dev, min_band, constant_ok);
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
  static OccCache occ_cache;
  static SmemOptIn smem_flag;
  if (int e = ensure_smem(kernel, smem, dev, smem_flag)) return e;
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
    // occupancy of this instantiation with this smem size
    const long long resident_warps =
        static_cast<long long>(cta_occupancy(kernel, smem, occ_cache, kCtaWarps * kWarp)) * kCtaWarps * dev.num_sms;
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

// Multi-channel band choice shared by the multi kernels: K >= 5 one full wave of resident warps (the
// K-1 prologue rows of extra bands cost more than the wave quantisation they remove --
// tools/multi_band_sweep.py: Table I CONV3/CONV5, configs[3]); K <= 4 the wave-quantisation cost model
// b* = argmin waves(b) * (ceil(Ho / b) + K - 1) (one band per tile whenever the (image group, F-block,
// column-block) groups alone exceed a wave had left Table I CONV11 at 1.15 waves: 946 -> 570 us).
// Returns n_bands padded so that the 4 warps of a CTA share (group, F-block); sets band_h.
template <int K>
int multi_bands(int Ho, int n_cb, long long groups, long long resident_ctas, int &band_h) {
  if (band_h <= 0 && K >= 5) {
    const long long resident_warps = resident_ctas * kCtaWarps;
    long long bands = resident_warps / (groups * n_cb);
    if (bands < 1) bands = 1;
    band_h = ceil_div(Ho, bands);
  } else if (band_h <= 0) {
    long long best_b = 1;
    double best = 1e300;
    const int bmax = Ho < 512 ? Ho : 512;
    for (int b = 1; b <= bmax; ++b) {
      const int h = ceil_div(Ho, b);
      const int nb = ceil_div(Ho, h);  // bands actually used with height h
      long long nbp = nb;
      while ((static_cast<long long>(n_cb) * nbp) % kCtaWarps) ++nbp;
      const long long ctas = groups * n_cb * nbp / kCtaWarps;
      const long long waves = (ctas + resident_ctas - 1) / resident_ctas;
      const double cost = static_cast<double>(waves) * (h + K - 1) * (1.0 + 1e-3 * (nbp - nb));
      if (cost < best - 1e-9) {
        best = cost;
        best_b = nb;
      }
    }
    band_h = ceil_div(Ho, best_b);
  }
  if (band_h > Ho) band_h = Ho;
  int n_bands = ceil_div(Ho, band_h);
  while ((static_cast<long long>(n_cb) * n_bands) % kCtaWarps) ++n_bands;
  return n_bands;
}

template <int K, int FB, int U, int SEG, int GUARDS, int PF, int MINB, bool ALIGNED, bool P2 = false>
int launch_multi2_k(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                    cudaStream_t stream, int band_h, const DevInfo &dev) {
  constexpr int KP = KCfg<K>::KP;
  constexpr int SEGS = kWarp / SEG;
  auto kernel = k_conv2d_multi2<K, FB, U, SEG, GUARDS, PF, MINB, ALIGNED, P2>;
  static OccCache occ_cache;
  static SmemOptIn smem_flag;
  const size_t ring = (PF >= 3) ? kCtaWarps * RowRing<K, U, SEG, PF>::kBytes : 0;
  // F-block filters (+ 16 bytes: the P2 layout C*K*K*FB floats may leave the ring 8-byte aligned only)
  const size_t fblock = P2 ? (static_cast<size_t>(C) * K * K * FB + 3) / 4 * 4 : static_cast<size_t>(C) * K * FB * KP;
  const size_t smem = fblock * sizeof(float) + ring;
  if (int e = ensure_smem(kernel, smem, dev, smem_flag)) return e;
  Multi2Args a;
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
  a.n_cb = ceil_div(a.Wo, 4 * SEG * U);
  a.n_fb = ceil_div(F, FB);
  a.n_groups = ceil_div(N, SEGS);
  a.aligned = (aligned16(in) && (W % 4 == 0)) ? 1 : 0;
  const long long resident_ctas =
      static_cast<long long>(cta_occupancy(kernel, smem, occ_cache, kCtaWarps * kWarp)) * dev.num_sms;
  const int n_bands = multi_bands<K>(a.Ho, a.n_cb, static_cast<long long>(a.n_groups) * a.n_fb, resident_ctas, band_h);
  a.band_h = band_h;
  a.n_bands = n_bands;
  a.n_tiles = static_cast<long long>(a.n_groups) * a.n_fb * n_bands * a.n_cb;
  const long long blocks = (a.n_tiles + kCtaWarps - 1) / kCtaWarps;
  if (blocks > 0x7fffffffLL) return CONV2D_ESHAPE;
  kernel<<<static_cast<unsigned>(blocks), kCtaWarps * kWarp, smem, stream>>>(a);
  return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
}


template <int K, int FB, int U, int SEG, int GUARDS, int PF, int MINB = (SEG == kWarp && K <= 3 && FB * U >= 8) ? 2 : 3,
          bool P2 = false>
int launch_multi2_v(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                    cudaStream_t stream, int band_h, const DevInfo &dev) {
  const bool aligned = aligned16(in) && (W % 4 == 0);
  if (!aligned)  // the misaligned-input instantiation (guarded scalar loads), its own register budget
    return launch_multi2_k<K, FB, U, SEG, GUARDS, PF, 2, false, P2>(in, N, C, H, W, filt, F, out, stream, band_h,
                                                                    dev);
  return launch_multi2_k<K, FB, U, SEG, GUARDS, PF, MINB, true, P2>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
}


// Filter-blocked multi-channel kernel (conv2d_mob.cuh). Warp-steps per warp L: the grid runs
// ceil(ctas / resident) waves of L steps each, so pick L minimising waves(L) * (L + 0.05) (the 0.05 step
// of F-block staging per CTA breaks ties towards fewer, longer CTAs). Returns CONV2D_ESHAPE when the
// F-block does not fit shared memory.
template <int K, int FB, int SEG, int EDGE, int MINB, bool PFL1 = false>
int launch_mob_k(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                 cudaStream_t stream, int L_req, const DevInfo &dev, long long *plan = nullptr) {
  constexpr int SEGS = kWarp / SEG;
  auto kernel = k_conv2d_mob<K, FB, SEG, EDGE, MINB, PFL1>;
  static OccCache occ_cache;
  static SmemOptIn smem_flag;
  const size_t smem = static_cast<size_t>(C) * K * K * FB * sizeof(float);
  if (int e = ensure_smem(kernel, smem, dev, smem_flag)) return e;
  MobArgs a;
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
  a.n_cb = ceil_div(a.Wo, kWideV * SEG);
  const long long units = static_cast<long long>(N) * a.Ho * a.n_cb;
  // 32-bit unit indices and channel-plane offsets in the kernel
  if (units + kCtaWarps * SEGS >= 0x7fffffffLL || static_cast<long long>(N) * C * H * W >= 0x7fffffffLL)
    return CONV2D_ESHAPE;  // (the round-1 kernel takes such tensors)
  a.units_img = a.Ho * a.n_cb;
  a.units = static_cast<int>(units);
  a.steps = (a.units + SEGS - 1) / SEGS;
  const int n_fb = ceil_div(F, FB);
  const uintptr_t ob = reinterpret_cast<uintptr_t>(out);
  a.ovec = ((ob & 15u) == 0 && a.Wo % 4 == 0) ? 2 : (((ob & 7u) == 0 && a.Wo % 2 == 0) ? 1 : 0);
  int L = L_req;
  const long long resident =
      static_cast<long long>(cta_occupancy(kernel, smem, occ_cache, kCtaWarps * kWarp)) * dev.num_sms;
  if (L <= 0) {
    // Only the smallest L of each wave count can be optimal (cost grows with L at fixed waves): for
    // w = 1 .. waves(L = 1), L_w = the smallest L whose grid fits in w waves. O(waves) host work per
    // call instead of O(steps); scanned with L ascending so ties keep the smallest L.
    const long long lmax = (a.steps + kCtaWarps - 1) / kCtaWarps;
    auto ctas_of = [&](long long l) { return static_cast<long long>(n_fb) * ((a.steps + kCtaWarps * l - 1) / (kCtaWarps * l)); };
    const long long w1 = (ctas_of(1) + resident - 1) / resident;
    double best = 1e300;
    L = 1;
    for (long long w = w1 < 65536 ? w1 : 65536; w >= 1; --w) {
      const long long m = w * resident / n_fb;  // CTAs per F-block that fit in w waves
      if (m < 1) continue;
      long long l = (a.steps + kCtaWarps * m - 1) / (kCtaWarps * m);
      if (l < 1) l = 1;
      if (l > lmax) l = lmax;
      const long long waves = (ctas_of(l) + resident - 1) / resident;
      const double cost = static_cast<double>(waves) * (static_cast<double>(l) + 0.05);
      if (cost < best - 1e-9) {
        best = cost;
        L = static_cast<int>(l);
      }
    }
  }
  a.L = L;
  a.n_fb = n_fb;
  a.ctas_fb = static_cast<int>((a.steps + static_cast<long long>(kCtaWarps) * L - 1) / (static_cast<long long>(kCtaWarps) * L));
  const long long blocks = static_cast<long long>(n_fb) * a.ctas_fb;
  if (blocks > 0x7fffffffLL) return CONV2D_ESHAPE;
  if (plan) {  // dry run: grid size and resident CTAs per wave
    plan[0] = blocks;
    plan[1] = resident;
    return CONV2D_OK;
  }
  kernel<<<static_cast<unsigned>(blocks), kCtaWarps * kWarp, smem, stream>>>(a);
  return cudaGetLastError() == cudaSuccess ? CONV2D_OK : CONV2D_ECUDA;
}

// segment width (lanes) of the filter-blocked kernel: the most lanes on valid columns (8*SEG-column
// units; a unit never straddles rows), ties to the wider segment. 32-lane segments are never strictly
// better than 16 (two 128-column units cover any row a 256-column unit covers) and are left to the
// tuning build.
inline int mob_seg(int Wo) {
  int best = 16;
  double bu = -1.0;
  for (int seg = 16; seg >= 4; seg /= 2) {
    const int span = kWideV * seg;
    const double u = double(Wo) / (double((Wo + span - 1) / span) * span);
    if (u > bu + 1e-9) {
      bu = u;
      best = seg;
    }
  }
  return best;
}

// aligned rows (W % 4 == 0, 16-byte base): clamped vector loads at MINB CTAs per SM; misaligned rows:
// the guarded scalar-load instantiation at MINB2 (its own register budget: 0 spills)
template <int K, int FB, int MINB, bool PFL1 = false, int MINB2 = (FB == 8 ? 2 : 3)>
int launch_mob(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
               cudaStream_t stream, int seg, int L_req, const DevInfo &dev, long long *plan = nullptr) {
  const bool aligned = aligned16(in) && (W % 4 == 0);
  if (seg <= 0) seg = mob_seg(W - K + 1);
#define C2D_MOB(S)                                                                                                \
  case S:                                                                                                         \
    return aligned ? launch_mob_k<K, FB, S, 1, MINB, PFL1>(in, N, C, H, W, filt, F, out, stream, L_req, dev, plan) \
                   : launch_mob_k<K, FB, S, 2, MINB2>(in, N, C, H, W, filt, F, out, stream, L_req, dev, plan);
  switch (seg) {
    C2D_MOB(4) C2D_MOB(8) C2D_MOB(16)
#ifdef C2D_TUNING
    C2D_MOB(32)
#endif
    default: return CONV2D_ESHAPE;
  }
#undef C2D_MOB
}

// The product multi-channel path (conv2d_mob.cuh). FB = 8 filters per lane at 3 CTAs per SM (168
// registers) for K <= 8, unless its grid fills less than 3/4 of one wave -- then FB = 4 (twice the
// CTAs, 4 CTAs per SM up to K = 6): Table I CONV4/6/7, tools/multi_variants.py, profiles/r02mob*.
// K >= 9: FB = 4 (ptxas spills FB = 8 there at 168 registers; 0 LDL/STL in every product kernel,
// tests/test_sass.py). band_h > 0: warp-steps per warp (explicit tiling; same bits). Returns
// CONV2D_ESHAPE when the F-block does not fit shared memory (caller falls back).
template <int K>
int launch_mob_auto(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                    cudaStream_t stream, int band_h, const DevInfo &dev) {
  constexpr int M4 = (K <= 6) ? 4 : 3;
  const int L = band_h > 0 ? band_h : 0;
  if constexpr (K <= 8) {
    long long plan[2] = {0, 0};
    const int e = launch_mob<K, 8, 3>(in, N, C, H, W, filt, F, out, stream, 0, L, dev, plan);
    if (e == CONV2D_OK && 4 * plan[0] >= 3 * plan[1]) {
      // K <= 4 with several channels: rows carry few FMAs and L1 misses (a new channel plane every
      // row) are exposed at one row of register prefetch -- an L1 prefetch two rows ahead: configs[2]
      // 25.6 -> 29.9 TFLOP/s, Table I C=3 K=3 layers +5-17%; C = 1 and K = 7 lose (profiles/r02_mob*)
      if constexpr (K <= 4)
        if (C >= 2) return launch_mob<K, 8, 3, true>(in, N, C, H, W, filt, F, out, stream, 0, L, dev);
      return launch_mob<K, 8, 3>(in, N, C, H, W, filt, F, out, stream, 0, L, dev);
    }
    if (e != CONV2D_OK && e != CONV2D_ESHAPE) return e;
  }
  return launch_mob<K, 4, M4>(in, N, C, H, W, filt, F, out, stream, 0, L, dev);
}

// fraction of a segment-row's lanes doing valid columns
inline double lane_use(int Wo, int span) { return double(Wo) / (double(ceil_div(Wo, span)) * span); }

template <int K>
int launch_multi(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                 cudaStream_t stream, int band_h, const DevInfo &dev) {
  // FB filters per warp (K*FB*4 accumulators); FBH = half of it (more warps, smaller loop body)
  constexpr int FB = (K <= 3) ? 8 : (K <= 7 ? 4 : 2);
  constexpr int FBH = (FB > 1) ? FB / 2 : 1;
  // the tuned default: FB = 8 filters per warp for K <= 3, half the register-limited FB above
  constexpr int FBD = (K <= 3) ? FB : FBH;
  constexpr int GUARDS = (K <= 5) ? 2 : 0;
  constexpr int KP = KCfg<K>::KP;
  const int Wo = W - K + 1;
  const int mv = tuning_mvariant();
  int rc = CONV2D_ESHAPE;
  // row prefetch: a 4-stage cp.async ring in shared memory for K >= 5; two entries in registers for
  // K <= 3, where a (row, channel) entry carries few FMAs and the ring's per-entry cost dominates
  constexpr int PF = (K <= 3) ? 2 : 4;
#define C2D_LM(FBB, SEGG) \
  launch_multi2_v<K, FBB, 1, SEGG, GUARDS, PF>(in, N, C, H, W, filt, F, out, stream, band_h, dev)
#ifdef C2D_TUNING
#define C2D_LM2(FBB, SEGG) \
  launch_multi2_v<K, FBB, 2, SEGG, GUARDS, PF>(in, N, C, H, W, filt, F, out, stream, band_h, dev)
  if (mv == 9) {  // the round-1 kernel
    constexpr int LFB = MultiCfg<K>::FB;
    const size_t lsmem = static_cast<size_t>(C) * K * LFB * KP * sizeof(float);
    if (lsmem <= static_cast<size_t>(dev.smem_optin))
      return launch_multi_fb<K, LFB>(in, N, C, H, W, filt, F, out, stream, band_h, dev, lsmem);
  }
  constexpr int FBQ = (FBH > 1) ? FBH / 2 : 1;
  if (mv == 5) return C2D_LM2(FBH, 16);
  if (mv == 6) return C2D_LM2(FBQ, 16);
  if (mv == 1) return C2D_LM(FB, 32);
  if (mv == 2) return C2D_LM(FB, 16);
  if (mv == 3) return C2D_LM(FBH, 32);
  if (mv == 4) return C2D_LM(FBH, 16);
  if (mv == 7) return (K > 3) ? C2D_LM(FBH, 8) : C2D_LM(FB, 8);
  // the pre-r02 register cap (3 CTAs per SM) for the FB = 8 kernels (spills at K <= 3)
  if (mv == 70) return launch_multi2_v<K, FB, 1, 16, GUARDS, PF, 3>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
  if (mv == 71) return launch_multi2_v<K, FB, 1, 8, GUARDS, PF, 3>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
  if (mv == 72) return launch_multi2_v<K, FB, 1, 32, GUARDS, PF, 3>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
  // paired FMA across filter pairs (row_step_multi_p2), the default FB: 16 / 8 / 32 lanes
  if constexpr (FBD % 2 == 0) {
    if (mv == 90) return launch_multi2_v<K, FBD, 1, 16, GUARDS, PF, 3, true>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
    if (mv == 91) return launch_multi2_v<K, FBD, 1, 8, GUARDS, PF, 3, true>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
    if (mv == 92) return launch_multi2_v<K, FBD, 1, 32, GUARDS, PF, 2, true>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
    if (mv == 93) return launch_multi2_v<K, FBD, 1, 16, GUARDS, PF, 2, true>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
  }
  // 8: the r02 default (k_conv2d_multi2: 4 columns per lane, K-slot ring, FB = 8 / 2 filters per warp).
  if (mv == 8) {
    // Tuned on B200 (tools/multi_variants.py): 16-lane segments (two images per warp) unless they waste
    // clearly more lanes than whole-warp rows -- more column blocks take the vector fast path and the
    // ragged edge is a smaller share.
    const bool seg16 = N >= 2 && lane_use(Wo, 64) >= lane_use(Wo, 128) - 0.05;
    // 8-lane segments (four images per warp, 32 columns each) for narrow layers: Table I's 8-26-column
    // outputs use 25-81% of the lanes instead of 12-41% (tools/multi_band_sweep.py)
    const bool seg8 = N >= 4 && Wo <= 32 && lane_use(Wo, 32) >= lane_use(Wo, 64) + 0.15;
    // K = 4..7 (two filters per warp): paired FMA across the filter pair (row_step_multi_p2, FFMA2) --
    // profiles/r02p_multi_p2.txt: configs[3] 42.6 vs 37.6 TFLOP/s, Table I K=5 layers +5-20%. K <= 3 (eight
    // filters per warp) keeps the scalar FMAs: its FFMA2 form spills at 3 CTAs per SM and loses at 2.
    constexpr bool P2 = (K >= 4 && K <= 7 && FBD % 2 == 0);
  #define C2D_LMP(SEGG) \
    launch_multi2_v<K, FBD, 1, SEGG, GUARDS, PF, (SEGG == kWarp && K <= 3 && FBD >= 8) ? 2 : 3, P2>( \
        in, N, C, H, W, filt, F, out, stream, band_h, dev)
    if (seg8)
      rc = C2D_LMP(8);
    else
      rc = seg16 ? C2D_LMP(16) : C2D_LMP(32);
  #undef C2D_LMP
    if (rc != CONV2D_ESHAPE) return rc;
  }
#undef C2D_LM2
  // filter-blocked kernel (conv2d_mob.cuh) at a fixed shape: 100 FB=8 (3 CTAs per SM, K <= 8) / 101 FB=4
  // with the automatic segment width; 102-105 FB=8 at 4/8/16/32-lane segments, 106-109 FB=4;
  // 112 FB=8 with the L1 prefetch two rows ahead (K <= 8)
  if (mv >= 100 && mv <= 112) {
    constexpr int M4 = (K <= 6) ? 4 : 3;
    const int segs[4] = {4, 8, 16, 32};
    if (mv == 101) return launch_mob<K, 4, M4>(in, N, C, H, W, filt, F, out, stream, 0, 0, dev);
    if (mv >= 106 && mv <= 109)
      return launch_mob<K, 4, M4>(in, N, C, H, W, filt, F, out, stream, segs[mv - 106], 0, dev);
    if constexpr (K <= 8) {
      if (mv == 100) return launch_mob<K, 8, 3>(in, N, C, H, W, filt, F, out, stream, 0, 0, dev);
      if (mv >= 102 && mv <= 105)
        return launch_mob<K, 8, 3>(in, N, C, H, W, filt, F, out, stream, segs[mv - 102], 0, dev);
      if (mv == 112) return launch_mob<K, 8, 3, true>(in, N, C, H, W, filt, F, out, stream, 0, 0, dev);
    }
    return CONV2D_EK;
  }
#endif
#undef C2D_LM
  // the filter-blocked kernel (conv2d_mob.cuh): profiles/r02_mob*, DESIGN.md section 5
  rc = launch_mob_auto<K>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
  if (rc != CONV2D_ESHAPE) return rc;
  // F-block does not fit shared memory: round-1 kernel with one filter per warp
  const size_t smem1 = static_cast<size_t>(C) * K * KP * sizeof(float);
  if (smem1 <= static_cast<size_t>(dev.smem_optin))
    return launch_multi_fb<K, 1>(in, N, C, H, W, filt, F, out, stream, band_h, dev, smem1);
  return CONV2D_ESHAPE;
}

}  // namespace

namespace c2d {

template <int K>
int single_entry(const float *in, int N, int H, int W, const float *filt, float *out, cudaStream_t stream,
                 int band_h, const DevInfo &dev, const float *in2, int H1, long long P, int Po) {
  const SingleGeom g{in, in2, N, H, W, H1, P, Po};
  return launch_single<K>(g, filt, out, stream, band_h, dev);
}

template <int K>
int multi_entry(const float *in, int N, int C, int H, int W, const float *filt, int F, float *out,
                cudaStream_t stream, int band_h, const DevInfo &dev) {
  return launch_multi<K>(in, N, C, H, W, filt, F, out, stream, band_h, dev);
}

template <int KH>
int rect_entry(const float *in, int H, int W, const float *filt, int KW, float *out, cudaStream_t stream,
               const DevInfo &dev) {
  switch (KW) {
#define C2D_RECT(KK) \
  case KK: return launch_rect_v<KH, KK>(in, H, W, filt, out, stream, dev);
    C2D_RECT(1) C2D_RECT(2) C2D_RECT(3) C2D_RECT(4) C2D_RECT(5) C2D_RECT(6) C2D_RECT(7) C2D_RECT(8)
    C2D_RECT(9) C2D_RECT(10) C2D_RECT(11) C2D_RECT(12) C2D_RECT(13) C2D_RECT(14) C2D_RECT(15)
#undef C2D_RECT
    default: return CONV2D_EK;
  }
}

}  // namespace c2d

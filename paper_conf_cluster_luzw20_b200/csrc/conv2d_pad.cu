// conv2d_pad.cu -- boundary and semantic variants of the single-channel call:
// 'same' output size with zero or replicate padding, and true (flipped-filter) convolution.
//
// Both reduce to the valid-mode, stride-1 cross-correlation the paper's kernels compute (PAPER.md
// P:83-85; R1/R2): true convolution is cross-correlation with the filter rotated
// by 180 degrees, and 'same' is the valid result on the image extended by K-1 rows and columns
// (top/left (K-1)/2, bottom/right K-1-(K-1)/2, the convention of torch.nn.functional.conv2d
// padding='same'). The rotation is a one-block kernel into the library's stream-ordered scratch
// pool. 'same' is computed as the interior -- one valid launch straight on the image, writing into
// the output with its row pitch (no extra pass over the image) -- plus four thin border strips whose
// slices of the extended image a small kernel materialises (16-byte row pitch) in the scratch pool,
// on a side stream concurrent with the interior.
// Every launch is the same per-K one-tile kernels (never the filter-row split), so the result is
// bitwise equal to the one-tile kernels on the fully padded image with the rotated filter.
#include <cstdint>
#include <mutex>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"
#include "common.h"

#ifndef C2D_PAD_INTERIOR_MAXK
#define C2D_PAD_INTERIOR_MAXK 9
#endif

namespace {

using namespace c2d;

// P[r][c] (r < Hp, c < P4*4) from in (H x W): padded column c maps to input column c - pl, row r to
// input row r - pt; out-of-range entries are 0 (ZERO) or the nearest edge element (REPLICATE);
// columns >= Wt (the pitch slack) are 0.
__global__ void k_pad_image(const float *__restrict__ in, int H, int W, float *__restrict__ P, int Hp, int Wt,
                            long long P4, int pt, int pl, int replicate, int er0, int ec0) {
  const long long total = static_cast<long long>(Hp) * P4;
  for (long long q = static_cast<long long>(blockIdx.x) * blockDim.x + threadIdx.x; q < total;
       q += static_cast<long long>(gridDim.x) * blockDim.x) {
    const int r = static_cast<int>(q / P4);
    const int c0 = static_cast<int>(q % P4) * 4;
    int ri = er0 + r - pt;  // (er0, ec0): this buffer's origin in the extended image
    const bool row_in = ri >= 0 && ri < H;
    if (replicate) ri = min(max(ri, 0), H - 1);
    float v[4];
#pragma unroll
    for (int t = 0; t < 4; ++t) {
      const int c = c0 + t;
      int ci = ec0 + c - pl;
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

// Border-strip side stream and its fork / join events: one set per (host thread, device), created on
// first use and kept, so concurrent callers on different threads never share a side stream.
struct SideSet {
  cudaStream_t stream = nullptr;
  cudaEvent_t fork = nullptr, join = nullptr;
  bool ok = false;
};
thread_local SideSet t_side[kMaxDevices];

SideSet *side_set(int dev) {
  if (dev < 0 || dev >= kMaxDevices) return nullptr;
  SideSet &ss = t_side[dev];
  if (!ss.ok) {
    if (cudaStreamCreateWithFlags(&ss.stream, cudaStreamNonBlocking) != cudaSuccess ||
        cudaEventCreateWithFlags(&ss.fork, cudaEventDisableTiming) != cudaSuccess ||
        cudaEventCreateWithFlags(&ss.join, cudaEventDisableTiming) != cudaSuccess) {
      (void)cudaGetLastError();
      return nullptr;
    }
    ss.ok = true;
  }
  return &ss;
}

bool capturing(cudaStream_t s) {
  cudaStreamCaptureStatus st = cudaStreamCaptureStatusNone;
  return cudaStreamIsCapturing(s, &st) == cudaSuccess && st != cudaStreamCaptureStatusNone;
}

int device_info(DevInfo *out) {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess) return CONV2D_ECUDA;
  out->id = dev;
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
  // One valid-mode launch of the per-K kernels: `src` (rows x cols, row pitch `pitch`) into `dst`
  // (output row pitch `po`). kBandNoSplit: the one-tile kernels everywhere in the padded call, so
  // interior and border outputs sum in the same order whatever the strip widths.
  auto conv_on = [&](cudaStream_t st, int band_flag, const float *src, int rows, int cols, long long pitch,
                     float *dst, int po) -> int {
    switch (K) {
#define C2D_CALL_PAD(KK) \
  case KK: return single_entry<KK>(src, 1, rows, cols, f_use, dst, st, band_flag, dev, src, rows, pitch, po);
      C2D_CALL_PAD(1) C2D_CALL_PAD(2) C2D_CALL_PAD(3) C2D_CALL_PAD(4) C2D_CALL_PAD(5) C2D_CALL_PAD(6)
      C2D_CALL_PAD(7) C2D_CALL_PAD(8) C2D_CALL_PAD(9) C2D_CALL_PAD(10) C2D_CALL_PAD(11) C2D_CALL_PAD(12)
      C2D_CALL_PAD(13) C2D_CALL_PAD(14) C2D_CALL_PAD(15)
#undef C2D_CALL_PAD
      default: return CONV2D_EK;
    }
  };
  auto conv = [&](const float *src, int rows, int cols, long long pitch, float *dst, int po) -> int {
    return conv_on(s, kBandNoSplit, src, rows, cols, pitch, dst, po);
  };
  if (!pad) {
    const int rc = conv(in, H, W, W, out, W - K + 1);
    if (f_rot) cudaFreeAsync(f_rot, s);
    return rc;
  }
  // 'same': out (H x W) = valid correlation of the extended image E ((H+K-1) x (W+K-1)). The interior
  // [pt, pt+H-K+1) x [pl, pl+W-K+1) reads only the image itself: one launch straight on `in`, writing
  // into `out` with row pitch W -- no extra pass over the image. The four border strips (top pt rows,
  // bottom pb rows, left pl / right pr columns of the rows between) each read a thin slice of E, which
  // k_pad_image materialises (16-byte pitch) in the scratch pool. Images smaller than the filter:
  // all of E at once.
  const int pt = (K - 1) / 2, pb = K - 1 - pt, pl = pt, pr = pb;
  struct Strip {
    int er0, ec0, rows, cols;  // slice of E
    long long out_off;         // first output element
  };
  Strip strips[5];
  int ns = 0;
  // The strips are latency-bound launches on images a few rows or columns wide: they run on a side
  // stream, concurrently with the interior (forked after the scratch allocation, joined before the
  // scratch is released), with the shared-memory filter so they never wait for the interior's use of
  // the constant slot. Same one-tile kernels, same bits. K < 9 (HBM-bound): 8192^2 K=3 'same' 0.197 ms
  // with the whole image padded -> 0.137 ms strips after the interior -> 0.128 ms concurrent strips.
  // K >= 9 (FMA-bound): the FMA-saturating interior leaves the strips no room, so the whole image is
  // padded instead (8192^2 K=15: 0.67 vs 0.68 ms).
  const bool interior = H >= K && W >= K && K < C2D_PAD_INTERIOR_MAXK;
  const int WE = W + K - 1;  // width of E
  if (!interior) {
    strips[ns++] = {0, 0, H + K - 1, WE, 0};
  } else {
    if (pt > 0) strips[ns++] = {0, 0, pt + K - 1, WE, 0};
    if (pb > 0) strips[ns++] = {H - pb, 0, pb + K - 1, WE, static_cast<long long>(H - pb) * W};
    if (pl > 0) strips[ns++] = {pt, 0, H, pl + K - 1, static_cast<long long>(pt) * W};
    if (pr > 0) strips[ns++] = {pt, W - pr, H, pr + K - 1, static_cast<long long>(pt) * W + W - pr};
  }
  long long off[5], total = 0;
  for (int t = 0; t < ns; ++t) {
    off[t] = total;
    const long long p4 = (strips[t].cols + 3) / 4 * 4;
    total += static_cast<long long>(strips[t].rows) * p4 + 4;  // +4: keeps every strip 16-byte aligned
  }
  float *scratch = nullptr;
  if (ns > 0 && scratch_alloc(reinterpret_cast<void **>(&scratch), static_cast<size_t>(total) * sizeof(float), s) !=
                    cudaSuccess) {
    if (f_rot) cudaFreeAsync(f_rot, s);
    return CONV2D_EALLOC;
  }
  int rc = CONV2D_OK;
  cudaStream_t ss = s;  // the strips' stream
  SideSet *side = nullptr;
  // Fork the strips onto this thread's side stream -- but not while `s` is being captured into a
  // graph: a side stream forked from a capturing stream joins that capture, so the strips stay on `s`.
  if (interior && ns > 0 && !capturing(s)) {
    side = side_set(dev.id);
    if (side && cudaEventRecord(side->fork, s) == cudaSuccess && cudaStreamWaitEvent(side->stream, side->fork, 0) == cudaSuccess)
      ss = side->stream;
  }
  // The interior first: the host enqueues the strips' ~10 small launches in tens of microseconds, and
  // enqueued after them the interior (the whole GPU's work) started that much later (8192^2 K=3
  // 'same': 0.20 ms vs 0.10 ms valid). The strips still overlap the interior's last wave.
  if (interior) rc = conv(in, H, W, W, out + static_cast<long long>(pt) * W + pl, W);
  for (int t = 0; t < ns && rc == CONV2D_OK; ++t) {
    const Strip &st = strips[t];
    const long long p4 = (st.cols + 3) / 4 * 4;
    float *buf = scratch + off[t];
    const long long quads = static_cast<long long>(st.rows) * (p4 / 4);
    long long blocks = (quads + 255) / 256;
    const long long cap = static_cast<long long>(dev.num_sms) * 8;
    if (blocks > cap) blocks = cap;
    k_pad_image<<<static_cast<unsigned>(blocks), 256, 0, ss>>>(in, H, W, buf, st.rows, st.cols, p4 / 4, pt, pl,
                                                               pad == CONV2D_PAD_REPLICATE ? 1 : 0, st.er0, st.ec0);
    if (cudaGetLastError() != cudaSuccess) rc = CONV2D_ECUDA;
    if (rc == CONV2D_OK)
      rc = conv_on(ss, ss == s ? kBandNoSplit : kBandSmemFilter, buf, st.rows, st.cols, p4, out + st.out_off, W);
  }
  if (ss != s) {  // join the strips back into the caller's stream (also on an error: nothing may dangle)
    if (cudaEventRecord(side->join, ss) != cudaSuccess || cudaStreamWaitEvent(s, side->join, 0) != cudaSuccess)
      rc = CONV2D_ECUDA;
  }
  if (scratch) cudaFreeAsync(scratch, s);
  if (f_rot) cudaFreeAsync(f_rot, s);
  return rc;
}

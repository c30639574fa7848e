// conv2d_host.cu -- conv2d_single_host: the end-to-end call on host buffers. A three-stage row-chunk
// pipeline (H2D copy of chunk i+1 | kernel of chunk i | D2H copy of chunk i-1) across two internal
// copy streams and the caller's stream, so PCIe traffic in both directions overlaps the kernels.
#include <algorithm>
#include <cstdint>
#include <mutex>
#include <vector>

#include <cuda_runtime.h>

#include "../../include/conv2d.h"
#include "common.h"

namespace {

using c2d::kMaxDevices;
constexpr int kEvents = 64;  // event ring (per device)

struct HostPipe {
  std::mutex mu;
  bool init = false;
  cudaStream_t s_in = nullptr, s_out = nullptr;
  cudaEvent_t ev[kEvents];
  int next = 0;
  cudaEvent_t get() {
    cudaEvent_t e = ev[next];
    next = (next + 1) % kEvents;
    return e;
  }
};
HostPipe g_pipe[kMaxDevices];

}  // namespace

extern "C" int conv2d_single_host(const float *in, int H, int W, const float *filt, int K, float *out, void *stream,
                                  int chunk_rows) {
  if (!in || !filt || !out) return CONV2D_ENULL;
  if (K < 1 || H < K || W < K) return K > CONV2D_MAX_K ? CONV2D_EK : CONV2D_ESHAPE;
  if (K > CONV2D_MAX_K) return CONV2D_EK;
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= kMaxDevices) return CONV2D_ECUDA;
  HostPipe &p = g_pipe[dev];
  {  // lazy init only; the copies and kernels below run without the lock (pageable copies block)
    std::lock_guard<std::mutex> lk(p.mu);
    if (!p.init) {
      if (cudaStreamCreateWithFlags(&p.s_in, cudaStreamNonBlocking) != cudaSuccess) return CONV2D_ECUDA;
      if (cudaStreamCreateWithFlags(&p.s_out, cudaStreamNonBlocking) != cudaSuccess) return CONV2D_ECUDA;
      for (int i = 0; i < kEvents; ++i)
        if (cudaEventCreateWithFlags(&p.ev[i], cudaEventDisableTiming) != cudaSuccess) return CONV2D_ECUDA;
      p.init = true;
    }
  }
  // an event of the ring (a stream wait captures the event's state when it is enqueued, so an event
  // re-recorded later by another call does not disturb an earlier wait)
  auto next_event = [&p]() {
    std::lock_guard<std::mutex> lk(p.mu);
    return p.get();
  };
  auto link = [&](cudaStream_t from, cudaStream_t to) {  // `to` waits for the work enqueued on `from`
    cudaEvent_t e = next_event();
    return cudaEventRecord(e, from) == cudaSuccess && cudaStreamWaitEvent(to, e, 0) == cudaSuccess;
  };
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  const int Ho = H - K + 1, Wo = W - K + 1;
  if (chunk_rows <= 0) chunk_rows = std::max(1, static_cast<int>((8ll << 20) / (4ll * W)));
  chunk_rows = std::min(chunk_rows, Ho);
  const size_t in_b = static_cast<size_t>(H) * W * sizeof(float);
  const size_t out_b = static_cast<size_t>(Ho) * Wo * sizeof(float);
  const size_t f_b = static_cast<size_t>(K) * K * sizeof(float);

  // everything starts after the work already on `stream`
  if (!link(s, p.s_in) || !link(s, p.s_out)) return CONV2D_ECUDA;

  void *d_buf = nullptr;
  const size_t in_pad = (in_b + 255) / 256 * 256, out_pad = (out_b + 255) / 256 * 256;
  if (c2d::scratch_alloc(&d_buf, in_pad + out_pad + f_b, p.s_in) != cudaSuccess) return CONV2D_EALLOC;
  float *d_in = static_cast<float *>(d_buf);
  float *d_out = reinterpret_cast<float *>(static_cast<char *>(d_buf) + in_pad);
  float *d_f = reinterpret_cast<float *>(static_cast<char *>(d_buf) + in_pad + out_pad);

  int rc = CONV2D_OK;
  if (cudaMemcpyAsync(d_f, filt, f_b, cudaMemcpyHostToDevice, p.s_in) != cudaSuccess) rc = CONV2D_ECUDA;
  int copied = 0;  // input rows already on the device
  for (int o0 = 0; o0 < Ho && rc == CONV2D_OK; o0 += chunk_rows) {
    const int rows = std::min(chunk_rows, Ho - o0);
    const int need = o0 + rows + K - 1;  // input rows [0, need) required for this chunk
    if (need > copied) {
      if (cudaMemcpyAsync(d_in + static_cast<size_t>(copied) * W, in + static_cast<size_t>(copied) * W,
                          static_cast<size_t>(need - copied) * W * sizeof(float), cudaMemcpyHostToDevice,
                          p.s_in) != cudaSuccess) {
        rc = CONV2D_ECUDA;
        break;
      }
      copied = need;
    }
    if (!link(p.s_in, s)) {
      rc = CONV2D_ECUDA;
      break;
    }
    rc = conv2d_single_ex(d_in + static_cast<size_t>(o0) * W, rows + K - 1, W, d_f, K,
                          d_out + static_cast<size_t>(o0) * Wo, s, 0);
    if (rc != CONV2D_OK) break;
    if (!link(s, p.s_out)) {
      rc = CONV2D_ECUDA;
      break;
    }
    if (cudaMemcpyAsync(out + static_cast<size_t>(o0) * Wo, d_out + static_cast<size_t>(o0) * Wo,
                        static_cast<size_t>(rows) * Wo * sizeof(float), cudaMemcpyDeviceToHost,
                        p.s_out) != cudaSuccess)
      rc = CONV2D_ECUDA;
  }
  // One exit path, also on errors: `stream` is ordered after everything enqueued on both copy
  // streams (nothing keeps writing into the caller's buffers unordered), then the scratch buffer is
  // released on `stream`.
  const bool joined = link(p.s_in, s) && link(p.s_out, s);
  if (cudaFreeAsync(d_buf, s) != cudaSuccess || !joined) return rc != CONV2D_OK ? rc : CONV2D_ECUDA;
  return rc;
}

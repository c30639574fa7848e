// FFMA vs FFMA2 (fma.rn.f32x2, sm_100) issue and FMA throughput with a uniform-register (UR) filter
// operand -- the operand form of the single-channel kernels. 8 independent accumulator chains per
// thread (pairs for FFMA2), a constant-bank coefficient per step.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/ffma2_rate tools/ubench/ffma2_rate.cu
#include <cstdio>
#include <cuda_runtime.h>

__constant__ float cf[64];

template <bool PAIR>
__global__ void __launch_bounds__(256) k(const float *in, float *out, int iters) {
  float a[16];
#pragma unroll
  for (int i = 0; i < 16; ++i) a[i] = in[threadIdx.x + i];
  float x0 = in[threadIdx.x + 100], x1 = in[threadIdx.x + 101];
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int j = 0; j < 32; ++j) {
      const float f = cf[j];
      if constexpr (PAIR) {
#pragma unroll
        for (int p = 0; p < 8; ++p) {
          unsigned long long d, xa, sa, fa;
          float2 xv = make_float2(x0, x1), sv = make_float2(a[2 * p], a[2 * p + 1]), fv = make_float2(f, f);
          xa = *reinterpret_cast<unsigned long long *>(&xv);
          sa = *reinterpret_cast<unsigned long long *>(&sv);
          fa = *reinterpret_cast<unsigned long long *>(&fv);
          asm volatile("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d) : "l"(xa), "l"(fa), "l"(sa));
          float2 r = *reinterpret_cast<float2 *>(&d);
          a[2 * p] = r.x;
          a[2 * p + 1] = r.y;
        }
      } else {
#pragma unroll
        for (int p = 0; p < 16; ++p) a[p] = fmaf((p & 1) ? x1 : x0, f, a[p]);
      }
    }
  }
  float s = 0.f;
#pragma unroll
  for (int i = 0; i < 16; ++i) s += a[i];
  out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

int main() {
  float h[64];
  for (int i = 0; i < 64; ++i) h[i] = 1.0f - 1e-6f * i;
  cudaMemcpyToSymbol(cf, h, sizeof(h));
  float *in, *out;
  cudaMalloc(&in, 1 << 20);
  cudaMalloc(&out, 148 * 8 * 256 * 4 * 4);
  cudaMemset(in, 0, 1 << 20);
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const int iters = 2000;
  for (int occ : {1, 2, 4, 8}) {
    const int blocks = sms * occ;
    for (int pair = 0; pair < 2; ++pair) {
      cudaEvent_t e0, e1;
      cudaEventCreate(&e0);
      cudaEventCreate(&e1);
      for (int rep = 0; rep < 2; ++rep) {
        cudaEventRecord(e0);
        if (pair) k<true><<<blocks, 256>>>(in, out, iters);
        else k<false><<<blocks, 256>>>(in, out, iters);
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
      }
      float ms = 0;
      cudaEventElapsedTime(&ms, e0, e1);
      const double fma = double(blocks) * 256 * iters * 32 * 16;
      printf("%s warps/SM %2d: %.3f ms, %.2f TFLOP/s fp32 (%.1f%% of 148x128x2x1.965G)\n", pair ? "FFMA2" : "FFMA ",
             occ * 8, ms, 2 * fma / ms / 1e9, 100.0 * 2 * fma / ms / 1e9 / 74.45);
    }
  }
  return 0;
}

// Does FFMA2 leave issue slots free? 16 FFMA2 (64 FMAs each) per step alone, then with 8 / 16 independent
// integer ops (IADD3 / LOP3, alu pipe) or 8 shuffles interleaved: if the FFMA2 pipe occupancy (2 cycles)
// hides the extra instructions, the time does not change.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/ffma2_dual tools/ubench/ffma2_dual.cu
#include <cstdio>
#include <cuda_runtime.h>

__constant__ float cf[64];

template <int NALU, bool SHFL, bool SCALAR>
__global__ void __launch_bounds__(256) k(const float *in, float *out, int iters) {
  float a[32];
#pragma unroll
  for (int i = 0; i < 32; ++i) a[i] = in[threadIdx.x + i];
  float x0 = in[threadIdx.x + 100], x1 = in[threadIdx.x + 101];
  unsigned u[16];
#pragma unroll
  for (int i = 0; i < 16; ++i) u[i] = threadIdx.x * (i + 1);
  float sh = x0;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int j = 0; j < 16; ++j) {
      const float f = cf[j];
      if constexpr (SCALAR) {
#pragma unroll
        for (int p = 0; p < 32; ++p) a[p] = fmaf((p & 1) ? x1 : x0, f, a[p]);
      } else {
#pragma unroll
        for (int p = 0; p < 16; ++p) {
          float2 r = __ffma2_rn(make_float2(x0, x1), make_float2(f, f), make_float2(a[2 * p], a[2 * p + 1]));
          a[2 * p] = r.x;
          a[2 * p + 1] = r.y;
        }
      }
#pragma unroll
      for (int q = 0; q < NALU; ++q) u[q] = (u[q] ^ (u[q] >> 3)) + 0x9E3779B9u;
      if constexpr (SHFL) {
#pragma unroll
        for (int q = 0; q < 8; ++q) sh = __shfl_sync(0xffffffffu, sh, (threadIdx.x + q + 1) & 31) + 1.0f;
      }
    }
  }
  float s = sh;
#pragma unroll
  for (int i = 0; i < 32; ++i) s += a[i];
  unsigned t = 0;
#pragma unroll
  for (int i = 0; i < 16; ++i) t ^= u[i];
  out[blockIdx.x * blockDim.x + threadIdx.x] = s + (float)t;
}

template <int NALU, bool SHFL, bool SCALAR>
void run(const char *name, int sms, const float *in, float *out) {
  const int iters = 1000, blocks = sms * 4;
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  for (int rep = 0; rep < 2; ++rep) {
    cudaEventRecord(e0);
    k<NALU, SHFL, SCALAR><<<blocks, 256>>>(in, out, iters);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
  }
  float ms = 0;
  cudaEventElapsedTime(&ms, e0, e1);
  const double fma = double(blocks) * 256 * iters * 16 * 32;
  printf("%-40s %.3f ms  %.2f TFLOP/s fp32 (%.1f%% of 74.45)\n", name, ms, 2 * fma / ms / 1e9,
         100.0 * 2 * fma / ms / 1e9 / 74.45);
}

int main() {
  float h[64];
  for (int i = 0; i < 64; ++i) h[i] = 1.0f - 1e-6f * i;
  cudaMemcpyToSymbol(cf, h, sizeof(h));
  float *in, *out;
  cudaMalloc(&in, 1 << 20);
  cudaMalloc(&out, 1 << 24);
  cudaMemset(in, 0, 1 << 20);
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  run<0, false, false>("FFMA2 x16 per step", sms, in, out);
  run<8, false, false>("FFMA2 x16 + 16 alu ops", sms, in, out);
  run<16, false, false>("FFMA2 x16 + 32 alu ops", sms, in, out);
  run<0, true, false>("FFMA2 x16 + 8 SHFL+FADD", sms, in, out);
  run<0, false, true>("FFMA x32 per step", sms, in, out);
  run<8, false, true>("FFMA x32 + 16 alu ops", sms, in, out);
  run<16, false, true>("FFMA x32 + 32 alu ops", sms, in, out);
  run<0, true, true>("FFMA x32 + 8 SHFL+FADD", sms, in, out);
  return 0;
}

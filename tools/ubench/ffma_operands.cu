// Micro-benchmark: FFMA throughput on sm_100a by operand form (3 registers / constant bank /
// immediate / shared-memory-fed register), the question behind the filter-supply design (DESIGN.md a4).
#include <cstdio>
#include <cuda_runtime.h>

__constant__ float c_f[64];

template <int MODE>
__global__ void __launch_bounds__(256) k(float *out, const float *fin, int iters) {
  __shared__ float sf[64];
  if (threadIdx.x < 64) sf[threadIdx.x] = fin[threadIdx.x];
  __syncthreads();
  float f[16];
#pragma unroll
  for (int j = 0; j < 16; ++j) f[j] = fin[j + (threadIdx.x & 1)];
  float acc[8], w[8];
#pragma unroll
  for (int v = 0; v < 8; ++v) { acc[v] = threadIdx.x * 1e-3f + v; w[v] = fin[32 + v]; }
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int j = 0; j < 16; ++j) {
      float fj;
      if (MODE == 0) fj = f[j];
      else if (MODE == 1) fj = c_f[j];
      else if (MODE == 2) fj = 1.0001f + j * 1e-5f;
      else { fj = sf[j + (it & 1)]; }
#pragma unroll
      for (int v = 0; v < 8; ++v) acc[v] = fmaf(acc[v], fj, w[v]);
    }
  }
  float s = 0;
#pragma unroll
  for (int v = 0; v < 8; ++v) s += acc[v];
  out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

int main() {
  float *out, *fin;
  cudaMalloc(&out, 148 * 8 * 256 * 4 * 4);
  cudaMalloc(&fin, 1024);
  cudaMemset(fin, 0, 1024);
  float h[64];
  for (int i = 0; i < 64; ++i) h[i] = 0.999f;
  cudaMemcpyToSymbol(c_f, h, sizeof(h));
  cudaMemcpy(fin, h, sizeof(h), cudaMemcpyHostToDevice);
  const int iters = 4096;
  const char *names[4] = {"3-reg", "const-bank", "immediate", "smem->reg"};
  for (int mode = 0; mode < 4; ++mode) {
    for (int occ : {4, 8}) {
      dim3 grid(148 * occ), block(256);
      cudaEvent_t e0, e1;
      cudaEventCreate(&e0);
      cudaEventCreate(&e1);
      auto launch = [&] {
        if (mode == 0) k<0><<<grid, block>>>(out, fin, iters);
        if (mode == 1) k<1><<<grid, block>>>(out, fin, iters);
        if (mode == 2) k<2><<<grid, block>>>(out, fin, iters);
        if (mode == 3) k<3><<<grid, block>>>(out, fin, iters);
      };
      launch();
      cudaEventRecord(e0);
      launch();
      cudaEventRecord(e1);
      cudaEventSynchronize(e1);
      float ms;
      cudaEventElapsedTime(&ms, e0, e1);
      double flops = 2.0 * grid.x * block.x * (double)iters * 16 * 8;
      printf("%-10s warps/SM=%2d: %.2f TFLOP/s\n", names[mode], occ * 8, flops / ms / 1e9);
    }
  }
  return 0;
}

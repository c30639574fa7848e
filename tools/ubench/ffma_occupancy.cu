// FFMA throughput vs warps per SM and independent chains per thread (sm_100a), 3-register form.
#include <cstdio>
#include <cuda_runtime.h>

template <int CH>
__global__ void __launch_bounds__(128) k(float *out, const float *fin, int iters) {
  float f[16];
#pragma unroll
  for (int j = 0; j < 16; ++j) f[j] = fin[j + (threadIdx.x & 1)];
  float acc[CH], w[CH];
#pragma unroll
  for (int v = 0; v < CH; ++v) { acc[v] = threadIdx.x * 1e-3f + v; w[v] = fin[32 + v]; }
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int j = 0; j < 16; ++j)
#pragma unroll
      for (int v = 0; v < CH; ++v) acc[v] = fmaf(acc[v], f[j], w[v]);
  }
  float s = 0;
#pragma unroll
  for (int v = 0; v < CH; ++v) s += acc[v];
  out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

template <int CH>
void run(float *out, float *fin) {
  for (int ctas : {1, 2, 3, 4, 6, 8}) {
    dim3 grid(148 * ctas), block(128);
    int iters = 4096 * 8 / CH;
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    k<CH><<<grid, block>>>(out, fin, iters);
    cudaEventRecord(e0);
    k<CH><<<grid, block>>>(out, fin, iters);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    double flops = 2.0 * grid.x * block.x * (double)iters * 16 * CH;
    printf("chains=%2d warps/SM=%2d: %.2f TFLOP/s\n", CH, ctas * 4, flops / ms / 1e9);
  }
}

int main() {
  float *out, *fin;
  cudaMalloc(&out, 148 * 8 * 128 * 4);
  cudaMalloc(&fin, 1024);
  float h[64];
  for (int i = 0; i < 64; ++i) h[i] = 0.999f;
  cudaMemcpy(fin, h, sizeof(h), cudaMemcpyHostToDevice);
  run<4>(out, fin);
  run<8>(out, fin);
  run<16>(out, fin);
  return 0;
}

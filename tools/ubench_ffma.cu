// Microbenchmark: FP32 FMA issue throughput on sm_100a for the operand forms the
// convolution kernels can use: weight in a register, weight in the constant bank
// (kernel parameter), and packed FFMA2 (fma.rn.f32x2). Not part of the product.
#include <cstdio>
#include <cuda_runtime.h>
struct W { float k[32]; };
struct W2 { float2 k[32]; };
#define NCH 8
__global__ void __launch_bounds__(256) ffma_const(float* out, int iters, const __grid_constant__ W w) {
  float a[NCH], x[NCH];
  #pragma unroll
  for (int c = 0; c < NCH; ++c) { a[c] = threadIdx.x * 1e-7f + c; x[c] = 1.0f + (threadIdx.x + c) * 1e-3f; }
  for (int it = 0; it < iters; ++it) {
    #pragma unroll
    for (int j = 0; j < 16; ++j)
      #pragma unroll
      for (int c = 0; c < NCH; ++c) a[c] = fmaf(x[c], w.k[j], a[c]);
  }
  float s = 0; for (int c = 0; c < NCH; ++c) s += a[c];
  if (s == 12345.f) out[threadIdx.x] = s;
}
__global__ void __launch_bounds__(256) ffma_reg(float* out, int iters, const float* wk) {
  float a[NCH], x[NCH], k[16];
  #pragma unroll
  for (int j = 0; j < 16; ++j) k[j] = wk[(j + threadIdx.x) & 15];
  #pragma unroll
  for (int c = 0; c < NCH; ++c) { a[c] = threadIdx.x * 1e-7f + c; x[c] = 1.0f + (threadIdx.x + c) * 1e-3f; }
  for (int it = 0; it < iters; ++it) {
    #pragma unroll
    for (int j = 0; j < 16; ++j)
      #pragma unroll
      for (int c = 0; c < NCH; ++c) a[c] = fmaf(x[c], k[j], a[c]);
  }
  float s = 0; for (int c = 0; c < NCH; ++c) s += a[c];
  if (s == 12345.f) out[threadIdx.x] = s;
}
__device__ __forceinline__ float2 ffma2(float2 a, float2 b, float2 c) {
  unsigned long long ra = *reinterpret_cast<unsigned long long*>(&a), rb = *reinterpret_cast<unsigned long long*>(&b),
                     rc = *reinterpret_cast<unsigned long long*>(&c), rd;
  asm("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(rd) : "l"(ra), "l"(rb), "l"(rc));
  return *reinterpret_cast<float2*>(&rd);
}
__global__ void __launch_bounds__(256) ffma2_const(float* out, int iters, const __grid_constant__ W2 w) {
  float2 a[NCH / 2], x[NCH / 2];
  #pragma unroll
  for (int c = 0; c < NCH / 2; ++c) { a[c] = make_float2(threadIdx.x * 1e-7f + c, c); x[c] = make_float2(1.0f + (threadIdx.x + c) * 1e-3f, threadIdx.y + 1.f); }
  for (int it = 0; it < iters; ++it) {
    #pragma unroll
    for (int j = 0; j < 16; ++j)
      #pragma unroll
      for (int c = 0; c < NCH / 2; ++c) a[c] = ffma2(x[c], w.k[j], a[c]);
  }
  float s = 0; for (int c = 0; c < NCH / 2; ++c) s += a[c].x + a[c].y;
  if (s == 12345.f) out[threadIdx.x] = s;
}
__global__ void __launch_bounds__(256) ffma2_reg(float* out, int iters, const float2* wk) {
  float2 a[NCH / 2], x[NCH / 2], k[16];
  #pragma unroll
  for (int j = 0; j < 16; ++j) k[j] = wk[(j + threadIdx.x) & 15];
  #pragma unroll
  for (int c = 0; c < NCH / 2; ++c) { a[c] = make_float2(threadIdx.x * 1e-7f + c, c); x[c] = make_float2(1.0f + (threadIdx.x + c) * 1e-3f, threadIdx.y + 1.f); }
  for (int it = 0; it < iters; ++it) {
    #pragma unroll
    for (int j = 0; j < 16; ++j)
      #pragma unroll
      for (int c = 0; c < NCH / 2; ++c) a[c] = ffma2(x[c], k[j], a[c]);
  }
  float s = 0; for (int c = 0; c < NCH / 2; ++c) s += a[c].x + a[c].y;
  if (s == 12345.f) out[threadIdx.x] = s;
}
int main() {
  int dev = 0; cudaDeviceProp p; cudaGetDeviceProperties(&p, dev);
  int clk = 0; cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, dev);
  printf("device %s SMs %d l2 %d MB smemOptin %zu clock(kHz) %d\n", p.name, p.multiProcessorCount, p.l2CacheSize >> 20, p.sharedMemPerBlockOptin, clk);
  float* out; cudaMalloc(&out, 4096); float* wk; cudaMalloc(&wk, 4096); cudaMemset(wk, 0, 4096);
  W w; W2 w2; for (int i = 0; i < 32; ++i) { w.k[i] = 0.5f + i * 1e-3f; w2.k[i] = make_float2(w.k[i], w.k[i]); }
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  int iters = 4096;
  for (int blocksPerSM : {1, 2, 4, 8}) {
    int grid = p.multiProcessorCount * blocksPerSM;
    double fmas = (double)grid * 256 * iters * 16 * NCH;
    for (int v = 0; v < 4; ++v) {
      float best = 1e30f;
      for (int rep = 0; rep < 5; ++rep) {
        cudaEventRecord(e0);
        if (v == 0) ffma_reg<<<grid, 256>>>(out, iters, wk);
        if (v == 1) ffma_const<<<grid, 256>>>(out, iters, w);
        if (v == 2) ffma2_reg<<<grid, 256>>>(out, iters, (const float2*)wk);
        if (v == 3) ffma2_const<<<grid, 256>>>(out, iters, w2);
        cudaEventRecord(e1); cudaEventSynchronize(e1);
        float ms; cudaEventElapsedTime(&ms, e0, e1); if (ms < best) best = ms;
      }
      const char* nm[] = {"ffma_reg", "ffma_const", "ffma2_reg", "ffma2_const"};
      double tf = fmas / (best * 1e-3) / 1e12;
      printf("%-12s warps/SM %2d : %.3f ms  %.2f T FMA/s  = %.1f FMA/clk/SM @1965MHz\n", nm[v], blocksPerSM * 8, best, tf,
             tf * 1e12 / (p.multiProcessorCount * 1.965e9));
    }
  }
  printf("err: %s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}

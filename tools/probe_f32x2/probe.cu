// Throughput probe: scalar FADD vs packed FADD2 (add.rn.f32x2, sm_100a) -- issue rate and
// FP32 lanes per SM-cycle, 8 independent chains per thread.
#include <cstdio>
#include <cuda_runtime.h>
typedef unsigned long long u64;
__device__ __forceinline__ u64 add2(u64 a, u64 b) { u64 d; asm volatile("add.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b)); return d; }
__global__ void k_scalar(float* out, int iters, float s) {
  float a[8];
#pragma unroll
  for (int i = 0; i < 8; ++i) a[i] = threadIdx.x * 0.001f + i;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < 8; ++i) a[i] = __fadd_rn(a[i], s);
  }
  float r = 0; for (int i = 0; i < 8; ++i) r += a[i];
  out[blockIdx.x * blockDim.x + threadIdx.x] = r;
}
__global__ void k_packed(float* out, int iters, float s) {
  u64 a[8];
  float2 sv = make_float2(s, s); u64 s2 = *reinterpret_cast<u64*>(&sv);
#pragma unroll
  for (int i = 0; i < 8; ++i) { float2 v = make_float2(threadIdx.x * 0.001f + i, i + 0.5f); a[i] = *reinterpret_cast<u64*>(&v); }
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < 8; ++i) a[i] = add2(a[i], s2);
  }
  float r = 0; for (int i = 0; i < 8; ++i) { float2 v = *reinterpret_cast<float2*>(&a[i]); r += v.x + v.y; }
  out[blockIdx.x * blockDim.x + threadIdx.x] = r;
}
int main() {
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  float* out; cudaMalloc(&out, sms * 8 * 1024 * sizeof(float));
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  const int iters = 20000;
  for (int threads : {256, 512, 1024}) {
    for (int pk = 0; pk < 2; ++pk) {
      for (int rep = 0; rep < 2; ++rep) {
        cudaEventRecord(e0);
        if (pk) k_packed<<<sms * 2, threads>>>(out, iters, 1e-7f); else k_scalar<<<sms * 2, threads>>>(out, iters, 1e-7f);
        cudaEventRecord(e1); cudaEventSynchronize(e1);
        float ms; cudaEventElapsedTime(&ms, e0, e1);
        double insts = (double)sms * 2 * threads * iters * 8;   // thread-instructions
        double flops = insts * (pk ? 2 : 1);
        if (rep) printf("%s threads/CTA=%d: %.3f ms, %.2f T thread-instr/s, %.2f T FP32 adds/s\n", pk ? "FADD2" : "FADD ", threads, ms, insts / ms / 1e9, flops / ms / 1e9);
      }
    }
  }
  return 0;
}

// Probe: does a 3-D TMA tile load accept a shared-memory destination that is only 16-B
// (not 128-B) aligned?  Loads the same box to offsets 0, 16, 32, 64 and compares.
#include <cuda.h>
#include <cudaTypedefs.h>
#include <cstdio>
#include <cstdint>
__device__ __forceinline__ uint32_t su(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__global__ void k(const __grid_constant__ CUtensorMap m, float* out, int off) {
  __shared__ __align__(1024) float tile[4096];
  __shared__ __align__(8) uint64_t bar;
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su(&bar)));
    asm volatile("fence.mbarrier_init.release.cluster;");
  }
  __syncthreads();
  float* dst = tile + off / 4;
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su(&bar)), "r"(8 * 10 * 3 * 4));
    asm volatile("cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];"
                 ::"r"(su(dst)), "l"(reinterpret_cast<uint64_t>(&m)), "r"(4), "r"(2), "r"(1), "r"(su(&bar)) : "memory");
  }
  asm volatile("{\n.reg .pred P1;\nW:\nmbarrier.try_wait.parity.shared::cta.b64 P1, [%0], 0;\n@!P1 bra W;\n}" ::"r"(su(&bar)));
  for (int i = threadIdx.x; i < 240; i += blockDim.x) out[i] = dst[i];
}
int main() {
  const int N0 = 8, N1 = 16, N2 = 32;
  float* g; cudaMalloc(&g, sizeof(float) * N0 * N1 * N2);
  float h[N0 * N1 * N2];
  for (int i = 0; i < N0 * N1 * N2; ++i) h[i] = (float)i;
  cudaMemcpy(g, h, sizeof(h), cudaMemcpyHostToDevice);
  void* fnp; cudaDriverEntryPointQueryResult q;
  cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fnp, cudaEnableDefault, &q);
  auto fn = (PFN_cuTensorMapEncodeTiled_v12000)fnp;
  CUtensorMap m;
  cuuint64_t dims[3] = {N2, N1, N0}, strides[2] = {N2 * 4, N1 * N2 * 4};
  cuuint32_t box[3] = {8, 10, 3}, es[3] = {1, 1, 1};
  fn(&m, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, g, dims, strides, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
     CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_NONE, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  float* d; cudaMalloc(&d, 240 * 4);
  for (int off : {0, 16, 32, 64}) {
    cudaMemset(d, 0, 240 * 4);
    k<<<1, 128>>>(m, d, off);
    cudaError_t e = cudaDeviceSynchronize();
    float r[240];
    cudaMemcpy(r, d, sizeof(r), cudaMemcpyDeviceToHost);
    int bad = 0;
    for (int z = 0; z < 3; ++z) for (int y = 0; y < 10; ++y) for (int x = 0; x < 8; ++x)
      bad += r[(z * 10 + y) * 8 + x] != h[((1 + z) * N1 + 2 + y) * N2 + 4 + x];
    printf("offset %d B: %s, %d mismatches\n", off, cudaGetErrorString(e), bad);
    if (e != cudaSuccess) return 1;
  }
  return 0;
}

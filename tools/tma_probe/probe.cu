// Minimal probe of a 3-D TMA tile load (debug tool).
#include <cuda.h>
#include <cudaTypedefs.h>
#include <cstdio>
#include <cstdint>
struct Maps { CUtensorMap m[2]; };
__device__ __forceinline__ uint32_t su(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__global__ void k(const __grid_constant__ Maps mp, float* out, int x, int y, int z, int which) {
  __shared__ __align__(128) float tile[18 * 36];
  __shared__ __align__(8) uint64_t bar;
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su(&bar)));
    asm volatile("fence.mbarrier_init.release.cluster;");
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su(&bar)), "r"(18 * 36 * 4));
    asm volatile("cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];"
                 ::"r"(su(tile)), "l"(reinterpret_cast<uint64_t>(&mp.m[which])), "r"(x), "r"(y), "r"(z), "r"(su(&bar)) : "memory");
  }
  asm volatile("{\n.reg .pred P1;\nW:\nmbarrier.try_wait.parity.shared::cta.b64 P1, [%0], 0;\n@!P1 bra W;\n}" ::"r"(su(&bar)));
  for (int i = threadIdx.x; i < 18 * 36; i += blockDim.x) out[i] = tile[i];
}
int main() {
  int N0 = 30, N1 = 37, N2 = 68;
  float* g; cudaMalloc(&g, sizeof(float) * N0 * N1 * N2);
  float* h = new float[N0 * N1 * N2];
  for (int i = 0; i < N0 * N1 * N2; ++i) h[i] = (float)i;
  cudaMemcpy(g, h, sizeof(float) * N0 * N1 * N2, cudaMemcpyHostToDevice);
  void* fnp; cudaDriverEntryPointQueryResult q;
  cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fnp, cudaEnableDefault, &q);
  auto fn = (PFN_cuTensorMapEncodeTiled_v12000)fnp;
  Maps mp;
  cuuint64_t dims[3] = {(cuuint64_t)N2, (cuuint64_t)N1, (cuuint64_t)N0};
  cuuint64_t str[2] = {(cuuint64_t)N2 * 4, (cuuint64_t)N1 * N2 * 4};
  cuuint32_t box[3] = {36, 18, 1}, es[3] = {1, 1, 1};
  for (int b = 0; b < 2; ++b) {
    CUresult r = fn(&mp.m[b], CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, g, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                    CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    printf("encode %d -> %d\n", b, (int)r);
  }
  float* o; cudaMalloc(&o, 18 * 36 * 4);
  int tests[6][3] = {{0, 0, 0}, {4, 3, 2}, {0, 3, 2}, {-4, -1, 1}, {8, 0, 0}, {1, 0, 0}};
  for (auto& t : tests) {
    k<<<1, 128>>>(mp, o, t[0], t[1], t[2], 1);
    cudaError_t e = cudaDeviceSynchronize();
    float r[18 * 36];
    cudaMemcpy(r, o, sizeof(r), cudaMemcpyDeviceToHost);
    printf("x=%d y=%d z=%d err=%s r[0]=%g r[37]=%g expect %g\n", t[0], t[1], t[2], cudaGetErrorString(e), r[0], r[37],
           (float)((t[2] * N1 + t[1] + 1) * N2 + t[0] + 1));
  }
  return 0;
}

// halo.cu -- the slab mode's halo staging copies (csrc/dist.cpp): the strided ghost slabs of a
// partition along a dimension > 0 (n_outer blocks of G lines, local_n lines apart) gathered into
// / scattered from contiguous NCCL buffers, optionally through a row list (only the outer rows
// whose state the next launch reads in that buffer).  One launch moves every region of one exchange (both
// ping-pong buffers, both sides) with 16-B loads and stores over a grid-stride loop -- four
// separate 2-D DMA copies per direction measured 0.36 ms per launch of heat-3D 1024^3 at 8 ranks
// (profiles/round2/dist_y), several times their HBM time.
#include <cstdint>

#include "launch.h"

namespace hexs {

namespace {

__global__ void __launch_bounds__(256) halo_copy_kernel(const __grid_constant__ HaloCopyArgs a) {
  // flattened (region, row, 16-B column) index space
  int64_t total = 0;
#pragma unroll 1
  for (int r = 0; r < a.n; ++r) total += (int64_t)a.reg[r].rows * (int64_t)(a.reg[r].width / 16);
  for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < total; e += (int64_t)gridDim.x * blockDim.x) {
    int64_t k = e;
    int r = 0;
    while (true) {
      const int64_t cnt = (int64_t)a.reg[r].rows * (int64_t)(a.reg[r].width / 16);
      if (k < cnt || r == a.n - 1) break;
      k -= cnt;
      ++r;
    }
    const HaloRegion& g = a.reg[r];
    const int64_t per = (int64_t)(g.width / 16);
    const int64_t row = k / per, col = k - row * per;
    const int64_t sr = g.src_rows ? g.src_rows[row] : row, dr = g.dst_rows ? g.dst_rows[row] : row;
    const uint4 v = *reinterpret_cast<const uint4*>(g.src + sr * (int64_t)g.spitch + col * 16);
    *reinterpret_cast<uint4*>(g.dst + dr * (int64_t)g.dpitch + col * 16) = v;
  }
}

}  // namespace

cudaError_t launch_halo_copy(const HaloCopyArgs& a, cudaStream_t s) {
  if (a.n <= 0) return cudaSuccess;
  if (a.n > kMaxHaloRegions) return cudaErrorInvalidValue;
  int64_t total = 0;
  for (int r = 0; r < a.n; ++r) {
    if (a.reg[r].width % 16 || a.reg[r].spitch % 16 || a.reg[r].dpitch % 16 ||
        (reinterpret_cast<uintptr_t>(a.reg[r].src) | reinterpret_cast<uintptr_t>(a.reg[r].dst)) % 16)
      return cudaErrorInvalidValue;
    total += (int64_t)a.reg[r].rows * (int64_t)(a.reg[r].width / 16);
  }
  int dev = 0, sms = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
  int64_t blocks = (total + 255) / 256;
  if (blocks > (int64_t)sms * 8) blocks = (int64_t)sms * 8;
  if (blocks < 1) blocks = 1;
  halo_copy_kernel<<<(int)blocks, 256, 0, s>>>(a);
  return cudaGetLastError();
}

}  // namespace hexs

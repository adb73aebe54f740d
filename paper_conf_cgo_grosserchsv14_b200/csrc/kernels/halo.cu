// halo.cu -- the slab mode's halo staging copies (csrc/dist.cpp): the strided ghost slabs of a
// partition along a dimension > 0 (n_outer blocks of G lines, local_n lines apart) gathered into
// / scattered from contiguous NCCL buffers, optionally through a row list (only the outer rows
// whose state the next launch reads in that buffer).  One launch moves every region of one exchange (both
// ping-pong buffers, both sides) with 16-B loads and stores over a grid-stride loop -- four
// separate 2-D DMA copies per direction measured 0.36 ms per launch of heat-3D 1024^3 at 8 ranks
// (profiles/round2/dist_y), several times their HBM time.
#include <cstdint>

#include <nccl.h>
#include <nccl_device.h>

#include "launch.h"

namespace hexs {

namespace {

__device__ __forceinline__ void copy_regions(const HaloCopyArgs& a) {
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

// Sender: copy into peer memory, then the last block to finish publishes seq to the neighbours.
__global__ void __launch_bounds__(256) halo_send_kernel(const __grid_constant__ HaloCopyArgs a,
                                                        const __grid_constant__ HaloSignal sig) {
  copy_regions(a);
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence_system();  // this block's peer stores before its completion count
    const unsigned int prev = atomicAdd(sig.done, 1u);
    if (prev == sig.done_base + gridDim.x - 1) {  // the last block: every block's stores are fenced
      __threadfence_system();
      for (int i = 0; i < sig.n; ++i)
        asm volatile("st.release.sys.global.b32 [%0], %1;" ::"l"(sig.flag[i]), "r"(sig.seq) : "memory");
    }
  }
}

// Receiver: one warp waits for the neighbours' sequence numbers (a single small CTA, so a
// co-scheduled peer kernel on the same device -- loopback mode -- always finds room); the
// scatter runs after it in stream order.
__global__ void __launch_bounds__(32) halo_wait_kernel(const __grid_constant__ HaloWait w) {
  if (threadIdx.x == 0) {
    for (int i = 0; i < w.n; ++i) {
      while (true) {
        int v;
        asm volatile("ld.acquire.sys.global.b32 %0, [%1];" : "=r"(v) : "l"(w.flag[i]) : "memory");
        if (v >= w.seq) break;
        __nanosleep(256);
      }
    }
    __threadfence_system();
  }
}

__global__ void halo_signal_kernel(int n, int* f0, int* f1, int seq) {
  __threadfence_system();
  if (n > 0) asm volatile("st.release.sys.global.b32 [%0], %1;" ::"l"(f0), "r"(seq) : "memory");
  if (n > 1) asm volatile("st.release.sys.global.b32 [%0], %1;" ::"l"(f1), "r"(seq) : "memory");
}

__global__ void __launch_bounds__(256) halo_copy_kernel(const __grid_constant__ HaloCopyArgs a) {
  copy_regions(a);
}

__global__ void peer_pointer_kernel(ncclWindow_t win, int peer, void** out) {
  out[0] = ncclGetPeerPointer(win, 0, peer);
}

}  // namespace

int halo_blocks() { return 4 * 148; }

cudaError_t launch_halo_send(const HaloCopyArgs& a, const HaloSignal& sig, int blocks, cudaStream_t s) {
  if (a.n > kMaxHaloRegions || sig.n > 2) return cudaErrorInvalidValue;
  halo_send_kernel<<<blocks, 256, 0, s>>>(a, sig);
  return cudaGetLastError();
}

cudaError_t launch_halo_recv(const HaloCopyArgs& a, const HaloWait& w, int blocks, cudaStream_t s) {
  if (a.n > kMaxHaloRegions || w.n > 2) return cudaErrorInvalidValue;
  halo_wait_kernel<<<1, 32, 0, s>>>(w);
  cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess || a.n == 0) return e;
  halo_copy_kernel<<<blocks, 256, 0, s>>>(a);
  return cudaGetLastError();
}

cudaError_t halo_peer_pointer(void* win, int peer, void** out, cudaStream_t s) {
  void** d = nullptr;
  cudaError_t e = cudaMallocAsync(reinterpret_cast<void**>(&d), sizeof(void*), s);
  if (e != cudaSuccess) return e;
  peer_pointer_kernel<<<1, 1, 0, s>>>(static_cast<ncclWindow_t>(win), peer, d);
  e = cudaGetLastError();
  if (e == cudaSuccess) e = cudaMemcpyAsync(out, d, sizeof(void*), cudaMemcpyDeviceToHost, s);
  if (e == cudaSuccess) e = cudaStreamSynchronize(s);
  cudaFreeAsync(d, s);
  return e;
}

cudaError_t launch_halo_signal(int n, int* const* flags, int seq, cudaStream_t s) {
  if (n <= 0) return cudaSuccess;
  if (n > 2) return cudaErrorInvalidValue;
  halo_signal_kernel<<<1, 1, 0, s>>>(n, flags[0], n > 1 ? flags[1] : nullptr, seq);
  return cudaGetLastError();
}

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

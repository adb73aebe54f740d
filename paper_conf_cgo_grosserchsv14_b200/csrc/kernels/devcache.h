// devcache.h -- per-device, thread-safe memo of host-side launch facts (dynamic shared
// memory attribute set, persistent grid size).  A process may drive plans on several
// devices (one plan per device); every such fact is a property of (kernel, device).
#pragma once
#include <mutex>

#include <cuda_runtime.h>

namespace hexs {

constexpr int kMaxDevices = 64;

// One value per device, computed once by `init()` on the current device (under a lock).
// `init` returns cudaSuccess and fills the value, or an error (not memoised).
template <typename V>
struct DeviceMemo {
  std::mutex mu;
  bool set[kMaxDevices] = {};
  V val[kMaxDevices] = {};

  template <typename F>
  cudaError_t get(V* out, F&& init) {
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return e;
    if (dev < 0 || dev >= kMaxDevices) return cudaErrorInvalidDevice;
    std::lock_guard<std::mutex> lk(mu);
    if (!set[dev]) {
      V v{};
      e = init(dev, &v);
      if (e != cudaSuccess) return e;
      val[dev] = v;
      set[dev] = true;
    }
    *out = val[dev];
    return cudaSuccess;
  }
};

}  // namespace hexs

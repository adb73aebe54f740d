// launch.h -- argument blocks and host-side launchers of the device kernels.
#pragma once
#include <cstdint>

#include <cuda_runtime.h>

namespace hexs {

constexpr int kMaxH = 64;

// General linear stencil (K_LINEAR): acc = c_0 A[p+d_0]; acc = acc + c_k A[p+d_k] (left to
// right), d_k the linear element offsets, over the interior [R, N-1-R] of every dimension.
constexpr int kMaxLin = 64;
struct LinearTerms {
  int n, R;
  int64_t delta[kMaxLin];
  double coef[kMaxLin];
};

// Generic hybrid kernel (Table 4 configuration (a): hybrid schedule, global memory only).
struct GenericArgs {
  void* f[3];      // ping-pong: f[0], f[1]; FDTD: ex, ey, hz (in place)
  int64_t N[3];    // extents slow -> fast (unused = 1)
  int64_t st[3];   // element strides
  int dims, hd, ncls;
  int cls[2], dcls[2], w[2];
  int64_t tau0;
  int a_lo, a_hi;
  int64_t S0_lo, row_off;
  int W;
  int64_t Slo[2], Shi[2];
  double k0, k1;
  int32_t lo[kMaxH], hi[kMaxH];
  // Wavefront execution of the classical tiles (wf = 1): persistent CTAs pull work items
  // (S0, S1, S2) in anti-diagonal order of (S1, S2); a tile starts once its predecessors
  // (S1-1, S2) and (S1, S2-1) of the same hexagon have published their completion flag.
  int wf;
  int64_t S0_hi;
  int* flags;                   // [nS0][n1][n2], zeroed before the launch
  unsigned long long* counter;  // work counter, zeroed before the launch
  LinearTerms lin;              // K_LINEAR: the access set and coefficients
};
cudaError_t launch_generic(int kind, int dtype, const GenericArgs& g, int grid, cudaStream_t s);
// Persistent grid size of the wavefront kernel (all CTAs co-resident).
int generic_wf_grid(int kind, int dtype);

// Naive one-step kernels (non-time-tiled comparator, K11).
struct NaiveArgs {
  const void* src;
  void* dst;
  void* f[3];  // FDTD fields
  int64_t N[3];
  double k0, k1;
  int stmt;    // FDTD statement 0 = ey, 1 = ex, 2 = hz
  LinearTerms lin;  // K_LINEAR
};
cudaError_t launch_naive(int kind, int dtype, int dims, const NaiveArgs& a, cudaStream_t s);

// Fast 2D register-wavefront hybrid kernel (jacobi / star5 / box9 / gradient2d).
struct Fast2DArgs {
  void* buf[2];
  int64_t N0, N1;
  int64_t tau0;
  int a_lo, a_hi, a_final;  // a_final: level whose outputs are level T_steps (-1: none)
  int64_t S0_lo, row_off;
  int W;
  double k0, k1;
};
cudaError_t launch_fast2d(int variant, const Fast2DArgs& a, int grid, cudaStream_t s);

// FDTD-2D fast kernel (kernels/fdtd.cu): one CTA per hexagon, j streamed through a
// shared-memory ring.
struct FdtdArgs {
  void* f[3];  // ex, ey, hz
  int64_t N0, N1;
  int64_t tau0;
  int a_lo, a_hi, a_final;
  int64_t S0_lo, row_off;
  int W;
  double k0, k1;
  int32_t lo[kMaxH], hi[kMaxH];  // hexagon rows per level
};
cudaError_t launch_fdtd(int variant, const FdtdArgs& a, int grid, cudaStream_t s);
size_t fdtd_smem_bytes(int dtype, int W);
int fdtd_ctas_per_sm();  // resident CTAs per SM the FDTD kernel is built for

// 3D fast kernel (kernels/hex3d.cu): persistent CTAs run the classical tiles of every
// hexagon of the launch as a tile-granular dependence wavefront, all levels of a tile in
// shared memory.
// A launch whose tiles a 3D launch reads (chained mode): its tile flags and tile geometry.
struct Fast3DPrev {
  const int* flags;  // nullptr: none
  const unsigned long long* done;  // its completed-tile counter (== its tile count: all complete)
  int64_t tau0, S0_lo, S0_hi, row_off, S1_lo, n1, S2_lo, n2;
};
struct Fast3DArgs {
  void* buf[2];
  int64_t N0, N1, N2;
  int64_t tau0;
  int a_lo, a_hi, a_final;
  int64_t S0_lo, S0_hi, row_off;
  int W, H, L, Q;          // box width, h, levels 2h+2, buffer rows (max hexagon rows + 2)
  int64_t S1_lo, n1, S2_lo, n2;
  double k0, k1;
  int* flags;                   // per tile completion flag, zeroed per launch
  unsigned long long* counter;  // work counter, zeroed per launch
  int32_t lo[kMaxH], hi[kMaxH];
  // Fused halo stores (multi-GPU slab mode along y, csrc/dist.cpp): every global store of a line
  // y in [mir_y0[s], mir_y0[s] + mir_G) is also written into neighbour s's mirror (peer memory),
  // laid out [buffer parity][z][y - mir_y0[s]][x]; mir[s] = nullptr: none.
  void* mir[2];
  int mir_y0[2];
  int mir_G;
  int mir_fence;  // 1: each thread that stored into a mirror fences at system scope before the tile's flag
  // Chained launches (single GPU): the launch may start while the previous two are still running
  // (programmatic dependent launch); before a tile's first fill its producer acquires the flags of
  // every tile of prev[0] (launch - 1) and prev[1] (launch - 2) that wrote a value it reads.
  Fast3DPrev prev[2];
  unsigned long long* done;  // this launch's completed-tile counter (chained mode; else nullptr)
  int pdl;  // 1: launched with programmatic stream serialization (and lets the next launch start early)
};
cudaError_t launch_fast3d(int variant, const Fast3DArgs& a, int grid, cudaStream_t s);

// Streaming 3D kernel (kernels/stream3d.cu): hexagons over (t, y), z streamed plane by plane
// (classical width 1, skew 1), x in strips of kStream3DNX (skew 4).  One CTA per (hexagon,
// strip), ticketed in (hexagon, strip) order; strips pass their right-edge quads through
// `scratch` (kStream3DRS steps deep) and publish per-step progress counters.
constexpr int kStream3DNX = 64;
constexpr int kStream3DRS = 32;
struct Stream3DArgs {
  void* buf[2];
  int64_t N0, N1, N2;
  int64_t tau0;
  int a_lo, a_hi, a_final;
  int64_t S0_lo, row_off;
  int W, L, RN;        // box width, levels 2h+2, hexagon rows 2h+w0+1
  int n_str, n_items;  // strips per hexagon, CTAs of the launch
  double k0, k1;
  int* progress;           // [n_items] completed steps, zeroed per launch
  unsigned int* ticket;    // CTA ticket counter, zeroed per launch
  float* scratch;          // [n_items][kStream3DRS][carry block]
};
cudaError_t launch_stream3d(int variant, const Stream3DArgs& a, cudaStream_t s);

// Table 4 ablation kernel (kernels/ablation.cu): one hybrid 3D phase kernel per memory strategy
// (a) global only .. (f) dynamic reuse, CTA 1 x 10 x 32 over classical tiles of 10 (y) x 32 (x).
enum { ABL_A = 0, ABL_B = 1, ABL_C = 2, ABL_D = 3, ABL_E = 4, ABL_F = 5 };
constexpr int kAblW1 = 10, kAblW2 = 32;
struct AblArgs {
  void* buf[2];
  int64_t N0, N1, N2;
  int64_t tau0;
  int a_lo, a_hi;
  int64_t S0_lo, S0_hi, row_off;
  int W;
  int64_t S1_lo, S2_lo;
  int n1, n2;            // y tiles (rows of the pipeline) and x tiles per row
  int ctrans1, ctrans2;  // classical translation offsets (tile bases B = S w + ctrans - a)
  int YB, XB, XP;        // shared box: y lines, x columns loaded, x pitch (64 = circular)
  double k0, k1;
  int* progress;               // [n1][nS0] completed x tiles per row, zeroed per launch
  unsigned int* counter;       // row ticket, zeroed per launch
  int32_t lo[kMaxH], hi[kMaxH];
};
cudaError_t launch_ablation(int cfg, int kind, const AblArgs& a, cudaStream_t s);
size_t ablation_smem_bytes(int cfg, int W, int YB, int XP);

// Slab-mode halo staging (kernels/halo.cu): up to kMaxHaloRegions strided 2-D copies in one
// launch (rows x width bytes, widths / pitches / pointers 16-B aligned).
constexpr int kMaxHaloRegions = 8;
struct HaloRegion {
  char* dst;
  const char* src;
  size_t dpitch, spitch, width, rows;
  const int* src_rows;  // optional row index lists (gather / scatter); nullptr = row i
  const int* dst_rows;
};
struct HaloCopyArgs {
  int n;
  HaloRegion reg[kMaxHaloRegions];
};
cudaError_t launch_halo_copy(const HaloCopyArgs& a, cudaStream_t s);

// Device-initiated halo exchange (kernels/halo.cu): the sender's kernel stores its halo lines
// straight into the neighbours' receive staging (peer memory over NVLink: an NCCL symmetric
// window's LSA pointers, or same-device pointers in loopback mode), and its last block publishes
// `seq` into the neighbours' flags (system-scope release); the receiver's kernel waits for the
// flags (acquire) and scatters its staging into its ghost lines.
struct HaloSignal {
  int n;                   // remote flags to publish
  int* flag[2];            // neighbour flag words (peer memory)
  unsigned int* done;      // this rank's block-completion counter (monotonic)
  unsigned int done_base;  // counter value before this launch
  int seq;
};
struct HaloWait {
  int n;                   // local flags to wait for
  const int* flag[2];
  int seq;
};
cudaError_t launch_halo_send(const HaloCopyArgs& a, const HaloSignal& sig, int blocks, cudaStream_t s);
cudaError_t launch_halo_recv(const HaloCopyArgs& a, const HaloWait& w, int blocks, cudaStream_t s);
int halo_blocks();  // grid of the send / receive kernels (fixed, so the completion counter is exact)
// publish seq into up to 2 flag words (peer memory) after a system-scope fence: everything this
// stream wrote before (e.g. a phase kernel's fused halo stores) is visible to the flags' readers
cudaError_t launch_halo_signal(int n, int* const* flags, int seq, cudaStream_t s);
// NCCL symmetric window: the peer's view of offset 0 of window `win` (a device-side LSA lookup)
cudaError_t halo_peer_pointer(void* win, int peer, void** out, cudaStream_t s);

}  // namespace hexs

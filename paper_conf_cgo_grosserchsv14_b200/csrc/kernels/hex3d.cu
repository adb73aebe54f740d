// hex3d.cu -- the specialised sm_100a phase kernel for 3D single-field stencils of radius 1
// (star3d7, gradient3d, box3d27) under the hybrid schedule: hexagonal over (t, z), classical
// parallelogram tiles over y and x (eq. (14)).
//
// Mapping:
//   * work item = one classical tile (S1, S2) of one hexagon S0 of the launch's (T, p): a
//     NY x NX (y, x) parallelogram over the hexagon's 2h+2 levels and rows z.  Skews: y by 1
//     per level (delta1_y = 1), x by 4 per level with a +1 tile translation (Sec. 4.2.3,
//     PAPER.md:755-763) so that every x-window this kernel moves starts on a 16-B boundary
//     (the TMA unit requires it; any skew >= delta1_x keeps eq. (14) valid -- reading R16);
//   * items run as a dependence WAVEFRONT at LEVEL granularity: level a of (S1, S2) needs
//     level a-1 of (S1-1, S2), (S1, S2-1), (S1-1, S2-1).  Persistent CTAs fetch items in
//     anti-diagonal order from an atomic counter; progress flags (levels done) are published
//     with st.release after the tile's carries are in global memory, so the ~26-51 hexagons
//     per phase of a 512^3 grid keep all 148 SMs busy -- the paper's mapping runs S1..Sn
//     sequentially inside one block;
//   * the tile's current level lives in shared memory (two level buffers: planes z x 18
//     lines x 40 columns); a thread owns 2 lines x 4 columns of one half of the rows and
//     sweeps z with a 3-plane register window (z-neighbours from registers, y/x neighbours
//     from LDS.128 + LDS.64);
//   * everything a tile reads from L2/HBM arrives by 3-D TMA tensor copies
//     (cp.async.bulk.tensor.3d, SASS UTMALDG) completing on one mbarrier per level buffer:
//     the In planes of level a+1 (the hexagon's slanted-edge inputs) one
//     level ahead, the carries (2 lines above / 5 columns left, produced by the predecessor
//     tiles in this launch) when their flags allow; out-of-grid box elements are zero-filled
//     by the TMA unit and never used;
//   * results leave from registers: the Out planes, the tile's last 2 lines and 5 columns
//     (its successors' carries) and the final level -- interleaved copy-out.
#include <cuda.h>
#include <cudaTypedefs.h>

#include <cstdint>

#include "../stencil_ops.cuh"
#include "launch.h"
#include "tma.cuh"

namespace hexs {
namespace fast3d {

constexpr int NY = kFast3DNY, NX = kFast3DNX;  // classical tile (y lines, x columns)
constexpr int NLP = NY / 2;                    // line pairs per tile
constexpr int NT = 2 * NLP * 8;                // 2 row groups x NLP line pairs x 8 column quads
constexpr int MINB = NY <= 8 ? 4 : 2;          // resident CTAs per SM (shared-memory bound)
constexpr int SIGMA = 4;                       // x skew per level
constexpr int CL = SIGMA + 1;                  // left carry columns (skew + stencil radius)
constexpr int LY = NY + 2;                     // buffer lines: 2 carry lines + NY
constexpr int SX = 40;                         // buffer columns: CL carry + NX window (+3), TMA box
constexpr int CW = 8;                          // carry-column box width (two 16-B groups of fp32)
// plane pitch (elements), padded so every TMA destination is 128-B aligned
template <typename T> constexpr int PP = ((LY * SX * (int)sizeof(T) + 127) / 128 * 128) / (int)sizeof(T);
template <typename T> constexpr size_t smem_bytes(int Q) {
  return (size_t)2 * Q * PP<T> * sizeof(T) + (size_t)Q * NY * CW * sizeof(T) + 128;
}

struct Maps {
  CUtensorMap plane[2];  // box {SX, LY, 1}   per ping-pong buffer
  CUtensorMap cline[2];  // box {SX, 2, 1}
  CUtensorMap ccol[2];   // box {CW, NY, 1}
};

__device__ __forceinline__ int ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ long long gtimer() {
  long long t;
  asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
  return t;
}
constexpr int kTraceStride = 32;  // per item: [sm, start, prologue, (flag, data, done) per level]

__device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.expect_tx.relaxed.cta.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}
__device__ __forceinline__ void tma_3d(void* dst, const CUtensorMap* map, int x, int y, int z, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::"r"(
          smem_u32(dst)),
      "l"(reinterpret_cast<uint64_t>(map)), "r"(x), "r"(y), "r"(z), "r"(smem_u32(bar))
      : "memory");
}

template <typename T, int KIND>
__device__ __forceinline__ T apply(const T (&x)[3][3][3], const Coef<T>& k) {
  // x[dz][dy][dx], offsets -1..1
  if constexpr (KIND == K_STAR3D7)
    return star3d7<T>(x[1][1][1], x[1][0][1], x[1][2][1], x[1][1][0], x[1][1][2], x[0][1][1], x[2][1][1], k);
  else if constexpr (KIND == K_GRADIENT3D)
    return gradient3d<T>(x[1][1][1], x[1][0][1], x[1][2][1], x[1][1][0], x[1][1][2], x[0][1][1], x[2][1][1], k);
  else {
    T acc = x[0][0][0];
#pragma unroll
    for (int q = 1; q < 27; ++q) acc = acc + x[q / 9][(q / 3) % 3][q % 3];
    return k.k0 * acc;
  }
}

// Buffer conventions.  The input buffer of level a (level a-1 values) has its column 0 at
// x = X0 - 4a (16-B aligned) and its line 0 at y = Y0 - a - 1: columns [0, CL) and lines
// {0, 1} are carries, the tile's own level-(a-1) window sits at columns [CL, CL + NX) and
// lines [2, LY).  Level a's output window (x in [X0-4a+1, X0-4a+NX], y in [Y0-a, Y0-a+NY))
// is written into the other buffer in ITS convention (column = x - (X0 - 4(a+1)),
// line = y - (Y0 - a - 2)).  A thread (lp, xq) computes outputs x = X0-4a+1+4xq+j,
// y = Y0-a+2lp+i, whose inputs sit at input columns [4xq, 4xq+5] and lines [2lp, 2lp+3].
template <typename T, int KIND>
__global__ void __launch_bounds__(NT, MINB) fast3d_kernel(const __grid_constant__ Fast3DArgs g,
                                                       const __grid_constant__ Maps m) {
  extern __shared__ __align__(1024) unsigned char smem_raw[];  // dynamic base is 1024-B aligned
  __shared__ __align__(8) uint64_t mbar[2];
  __shared__ int64_t item_s[3];
  __shared__ int64_t trace_it_s;
  T* buf = reinterpret_cast<T*>(smem_raw);  // stays a shared-space pointer (LDS/STS, not generic LD/ST)
  T* side = buf + (size_t)2 * g.Q * PP<T>;  // [Q][NY][CW] landing area of the carry columns
  auto B = [&](int which, int q, int ly, int lx) -> T* {
    return buf + ((size_t)which * g.Q + q) * PP<T> + ly * SX + lx;
  };
  const Coef<T> cf{(T)g.k0, (T)g.k1};
  const int tid = threadIdx.x;
  const int zg = tid / (NLP * 8), lp = (tid >> 3) % NLP, xq = tid & 7;  // row group (= warp for NY=8), line pair, col quad
  const int64_t ns0 = g.S0_hi - g.S0_lo + 1;
  const int64_t n1 = g.n1, n2 = g.n2, n_items = ns0 * n1 * n2;
  const int64_t plane = g.N1 * g.N2;
  const uint32_t plane_bytes = LY * SX * sizeof(T), cline_bytes = 2 * SX * sizeof(T),
                 ccol_bytes = NY * CW * sizeof(T);
  if (tid == 0) {
    mbar_init(&mbar[0], 1);
    mbar_init(&mbar[1], 1);
    mbar_fence_init();
  }
  __syncthreads();
  uint32_t phase[2] = {0u, 0u};

  while (true) {
    if (tid == 0) {
      const int64_t it = (int64_t)atomicAdd(g.counter, 1ull);
      int64_t S0 = -1, q1 = 0, q2 = 0;
      if (it < n_items) {  // decode: anti-diagonal d = q1 + q2 (outer), then S0, then q1
        int64_t off = 0;
        for (int64_t d = 0; d < n1 + n2 - 1; ++d) {
          const int64_t lo1 = d - (n2 - 1) > 0 ? d - (n2 - 1) : 0;
          const int64_t hi1 = d < n1 - 1 ? d : n1 - 1;
          const int64_t pairs = hi1 - lo1 + 1;
          if (it < off + pairs * ns0) {
            const int64_t r = it - off;
            S0 = g.S0_lo + r / pairs;
            q1 = lo1 + r % pairs;
            q2 = d - q1;
            break;
          }
          off += pairs * ns0;
        }
      }
      item_s[0] = S0;
      item_s[1] = q1;
      item_s[2] = q2;
      if (g.trace && it < n_items) {
        unsigned smid;
        asm volatile("mov.u32 %0, %smid;" : "=r"(smid));
        g.trace[it * kTraceStride] = ((long long)smid << 32) | (long long)(q1 * 65536 + q2);
        g.trace[it * kTraceStride + 1] = gtimer();
        item_s[0] = S0;
      }
      trace_it_s = it;
    }
    __syncthreads();
    const int64_t S0 = item_s[0];
    if (S0 < 0) break;
    const int64_t q1 = item_s[1], q2 = item_s[2];
    const int64_t fbase = (S0 - g.S0_lo) * n1 * n2;
    int* my_flag = g.flags + fbase + q1 * n2 + q2;
    const int64_t i0 = S0 * g.W - g.row_off;  // z of local row b = 0 (buffer plane q = b + 1)
    const int64_t Y0 = (g.S1_lo + q1) * NY, X0 = (g.S2_lo + q2) * NX;

    // prologue: every input plane of the first level (produced by earlier launches)
    {
      const int a = g.a_lo, ib = a & 1;
      if (tid == 0) {
        fence_proxy_async_smem();
        const int qlo = g.lo[a], qhi = g.hi[a] + 2;
        mbar_arrive_expect_tx(&mbar[ib], plane_bytes * (qhi - qlo + 1));
        const CUtensorMap* mp = &m.plane[(g.tau0 + a) & 1];
        for (int q = qlo; q <= qhi; ++q)
          tma_3d(B(ib, q, 0, 0), mp, (int)(X0 - SIGMA * a), (int)(Y0 - a - 1), (int)(i0 + q - 1), &mbar[ib]);
      }
      mbar_wait_parity(&mbar[ib], phase[ib]);
      phase[ib] ^= 1u;
    }
    long long* tr = (g.trace && tid == 0) ? g.trace + trace_it_s * kTraceStride : nullptr;
    if (tr) tr[2] = gtimer();

    for (int a = g.a_lo; a <= g.a_hi; ++a) {
      const int tk = 3 + 3 * (a - g.a_lo);
      const int ib = a & 1, ob = (a + 1) & 1;
      if (a > g.a_lo) {
        const int plo = g.lo[a - 1], phi = g.hi[a - 1];  // rows computed at level a-1
        // (0) level-granular dependences, then the carries of level a (TMA)
        if (tid == 0) {
          const int need = a - g.a_lo;
          if (q1 > 0)
            while (ld_acquire(g.flags + fbase + (q1 - 1) * n2 + q2) < need) __nanosleep(20);
          if (q2 > 0)
            while (ld_acquire(g.flags + fbase + q1 * n2 + q2 - 1) < need) __nanosleep(20);
          if (q1 > 0 && q2 > 0)
            while (ld_acquire(g.flags + fbase + (q1 - 1) * n2 + q2 - 1) < need) __nanosleep(20);
          if (tr) tr[tk] = gtimer();
          fence_proxy_async_smem();
          mbar_arrive_expect_tx(&mbar[ib], (cline_bytes + ccol_bytes) * (phi - plo + 1));
          const int par = (int)((g.tau0 + a) & 1);
          const int xo = (int)(X0 - SIGMA * a);
          for (int q = plo + 1; q <= phi + 1; ++q) {
            const int z = (int)(i0 + q - 1);
            tma_3d(B(ib, q, 0, 0), &m.cline[par], xo, (int)(Y0 - a - 1), z, &mbar[ib]);
            tma_3d(side + (size_t)q * NY * CW, &m.ccol[par], xo, (int)(Y0 - a + 1), z, &mbar[ib]);
          }
        }
        mbar_wait_parity(&mbar[ib], phase[ib]);  // carries + the In planes issued at level a-1
        phase[ib] ^= 1u;
        if (tr) tr[tk + 1] = gtimer();
        // the CL carry columns of each computed plane into place
        const int nc = phi - plo + 1;
        for (int e = tid; e < nc * NY * CL; e += NT) {
          const int q = plo + 1 + e / (NY * CL), r = e % (NY * CL), l = r / CL, c = r % CL;
          *B(ib, q, 2 + l, c) = side[((size_t)q * NY + l) * CW + c];
        }
        __syncthreads();
      }
      // (1) one level ahead: the In planes of level a+1 (areas level a does not write)
      if (a < g.a_hi && tid == 0) {
        const int qlo = g.lo[a + 1], qhi = g.hi[a + 1] + 2;
        int n_in = 0;
        for (int q = qlo; q <= qhi; ++q)
          if (q - 1 < g.lo[a] || q - 1 > g.hi[a]) ++n_in;
        fence_proxy_async_smem();
        mbar_expect_tx(&mbar[ob], plane_bytes * n_in);
        const CUtensorMap* mp = &m.plane[(g.tau0 + a + 1) & 1];
        for (int q = qlo; q <= qhi; ++q)
          if (q - 1 < g.lo[a] || q - 1 > g.hi[a])
            tma_3d(B(ob, q, 0, 0), mp, (int)(X0 - SIGMA * (a + 1)), (int)(Y0 - a - 2), (int)(i0 + q - 1), &mbar[ob]);
      }

      // (2) compute level a: rows [lo, hi] in two groups, z-window rotated without copies
      const int rlo = g.lo[a], rhi = g.hi[a];
      const int mid = (rlo + rhi) >> 1;
      const int r0 = zg == 0 ? rlo : mid + 1, r1 = zg == 0 ? mid : rhi;
      const int64_t yb = Y0 - a + 2 * lp, xb = X0 - SIGMA * a + 1 + 4 * xq;  // output (0, 0)
      // per-output masks (bit i*4+j): interior in (y, x); successors' carry cells
      uint32_t vmask = 0, cmask = 0;
#pragma unroll
      for (int i = 0; i < 2; ++i)
#pragma unroll
        for (int j = 0; j < 4; ++j) {
          const bool ok = (yb + i >= 1) && (yb + i <= g.N1 - 2) && (xb + j >= 1) && (xb + j <= g.N2 - 2);
          const bool carry = (lp == NLP - 1) || (4 * xq + j >= NX - CL);
          vmask |= (ok ? 1u : 0u) << (i * 4 + j);
          cmask |= (ok && carry ? 1u : 0u) << (i * 4 + j);
        }
      T* dst = static_cast<T*>(g.buf[(g.tau0 + a + 1) & 1]);
      const bool fin = (a == g.a_final);

      auto load_plane = [&](int q, T (&w)[4][6]) {
#pragma unroll
        for (int l = 0; l < 4; ++l) {
          const T* p = B(ib, q, 2 * lp + l, 4 * xq);
          if constexpr (sizeof(T) == 4) {
            const float4 u = reinterpret_cast<const float4*>(p)[0];
            const float2 v = reinterpret_cast<const float2*>(p)[2];
            w[l][0] = u.x; w[l][1] = u.y; w[l][2] = u.z; w[l][3] = u.w; w[l][4] = v.x; w[l][5] = v.y;
          } else {
#pragma unroll
            for (int i = 0; i < 3; ++i) {
              const double2 u = reinterpret_cast<const double2*>(p)[i];
              w[l][2 * i] = u.x; w[l][2 * i + 1] = u.y;
            }
          }
        }
      };
      auto step = [&](int r, const T (&P)[4][6], const T (&C)[4][6], const T (&N)[4][6]) {
        const int64_t z = i0 + r;
        const bool zok = (z >= 1) && (z <= g.N0 - 2);
        const uint32_t okm = zok ? vmask : 0u;
        T out[2][4];
#pragma unroll
        for (int i = 0; i < 2; ++i)
#pragma unroll
          for (int j = 0; j < 4; ++j) {
            T x[3][3][3];
#pragma unroll
            for (int dy = 0; dy < 3; ++dy)
#pragma unroll
              for (int dx = 0; dx < 3; ++dx) {
                x[0][dy][dx] = P[i + dy][j + dx];
                x[1][dy][dx] = C[i + dy][j + dx];
                x[2][dy][dx] = N[i + dy][j + dx];
              }
            const T v = apply<T, KIND>(x, cf);
            out[i][j] = ((okm >> (i * 4 + j)) & 1u) ? v : x[1][1][1];
          }
        // into the output buffer: columns CL + 4xq + j (one scalar, one pair, one scalar)
#pragma unroll
        for (int i = 0; i < 2; ++i) {
          T* p = B(ob, r + 1, 2 + 2 * lp + i, CL + 4 * xq);
          p[0] = out[i][0];
          if constexpr (sizeof(T) == 4) reinterpret_cast<float2*>(p + 1)[0] = make_float2(out[i][1], out[i][2]);
          else { p[1] = out[i][1]; p[2] = out[i][2]; }
          p[3] = out[i][3];
        }
        // copy-out from registers: Out planes / final level in full, else the successors'
        // carries (the window's last 2 lines and last CL columns)
        bool full = fin;
        if (a == g.H) full = full || r == rlo || r == rhi;
        else if (a > g.H && a < g.L - 1) full = full || r <= rlo + 1 || r >= rhi - 1;
        else if (a == g.L - 1) full = true;
        const uint32_t sm_ = zok ? (full ? vmask : cmask) : 0u;
        if (sm_) {
          T* rp = dst + z * plane + yb * g.N2 + xb;
#pragma unroll
          for (int i = 0; i < 2; ++i)
#pragma unroll
            for (int j = 0; j < 4; ++j)
              if ((sm_ >> (i * 4 + j)) & 1u) rp[i * g.N2 + j] = out[i][j];
        }
      };

      if (r0 <= r1) {
        T wa[4][6], wb[4][6], wc[4][6];
        load_plane(r0, wa);      // plane of row r0 - 1
        load_plane(r0 + 1, wb);  // plane of row r0
        int r = r0;
        while (true) {
          if (r > r1) break;
          load_plane(r + 2, wc);
          step(r, wa, wb, wc);
          if (++r > r1) break;
          load_plane(r + 2, wa);
          step(r, wb, wc, wa);
          if (++r > r1) break;
          load_plane(r + 2, wb);
          step(r, wc, wa, wb);
          ++r;
        }
      }
      __syncthreads();  // level a complete in ob; every thread's stores of level a issued
      // st.release.gpu after the CTA barrier is cumulative over the barrier-ordered stores of
      // every thread of the CTA (PTX memory model), so no separate membar is needed
      if (tid == 0) st_release(my_flag, a - g.a_lo + 1);
      if (tr) tr[tk + 2] = gtimer();
    }
  }
}

static PFN_cuTensorMapEncodeTiled_v12000 get_encode() {
  static PFN_cuTensorMapEncodeTiled_v12000 fn = nullptr;
  if (!fn) {
    cudaDriverEntryPointQueryResult q;
    void* p = nullptr;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
  }
  return fn;
}

template <typename T>
static bool encode(CUtensorMap* map, void* base, const Fast3DArgs& a, uint32_t bx, uint32_t by) {
  auto fn = get_encode();
  if (!fn) return false;
  cuuint64_t dims[3] = {(cuuint64_t)a.N2, (cuuint64_t)a.N1, (cuuint64_t)a.N0};
  cuuint64_t strides[2] = {(cuuint64_t)a.N2 * sizeof(T), (cuuint64_t)a.N1 * a.N2 * sizeof(T)};
  cuuint32_t box[3] = {bx, by, 1};
  cuuint32_t es[3] = {1, 1, 1};
  const CUtensorMapDataType dt = sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64;
  return fn(map, dt, 3, base, dims, strides, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE,
            CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE) == CUDA_SUCCESS;
}

static long long* g_trace = nullptr;
static int64_t g_trace_launch = -1, g_launch_count = 0;

template <typename T, int KIND>
cudaError_t launch_t(const Fast3DArgs& a_in, cudaStream_t s) {
  Fast3DArgs a = a_in;
  a.trace = (g_trace && g_launch_count++ == g_trace_launch) ? g_trace : nullptr;
  static int grid = 0;
  static size_t attr_bytes = 0;
  const size_t smem = smem_bytes<T>(a.Q);
  if (smem > attr_bytes) {
    cudaError_t e = cudaFuncSetAttribute(fast3d_kernel<T, KIND>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    attr_bytes = smem;
    grid = 0;
  }
  if (grid == 0) {
    int dev = 0, sms = 0, per_sm = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, fast3d_kernel<T, KIND>, NT, smem);
    grid = sms * (per_sm > 0 ? per_sm : 1);
  }
  Maps m;
  for (int b = 0; b < 2; ++b) {
    if (!encode<T>(&m.plane[b], a.buf[b], a, SX, LY) || !encode<T>(&m.cline[b], a.buf[b], a, SX, 2) ||
        !encode<T>(&m.ccol[b], a.buf[b], a, CW, NY))
      return cudaErrorInvalidValue;
  }
  fast3d_kernel<T, KIND><<<grid, NT, smem, s>>>(a, m);
  return cudaGetLastError();
}

}  // namespace fast3d

void fast3d_set_trace(long long* dev_buf, int64_t launch_index) {
  fast3d::g_trace = dev_buf;
  fast3d::g_trace_launch = launch_index;
  fast3d::g_launch_count = 0;
}

size_t fast3d_smem_bytes(int dtype, int Q) {
  return dtype == 1 ? fast3d::smem_bytes<double>(Q) : fast3d::smem_bytes<float>(Q);
}

// variant id = kind * 2 + dtype for the 3D classes
cudaError_t launch_fast3d(int variant, const Fast3DArgs& a, int /*grid: persistent*/, cudaStream_t s) {
  switch (variant) {
    case K_STAR3D7 * 2: return fast3d::launch_t<float, K_STAR3D7>(a, s);
    case K_STAR3D7 * 2 + 1: return fast3d::launch_t<double, K_STAR3D7>(a, s);
    case K_GRADIENT3D * 2: return fast3d::launch_t<float, K_GRADIENT3D>(a, s);
    case K_GRADIENT3D * 2 + 1: return fast3d::launch_t<double, K_GRADIENT3D>(a, s);
    case K_BOX3D27 * 2: return fast3d::launch_t<float, K_BOX3D27>(a, s);
    case K_BOX3D27 * 2 + 1: return fast3d::launch_t<double, K_BOX3D27>(a, s);
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace hexs

// Debug hook (not part of include/stencil.h): trace one 3D launch's per-item timeline.
extern "C" void hexs_debug_fast3d_trace(void* dev_buf, int64_t launch_index) {
  hexs::fast3d_set_trace(static_cast<long long*>(dev_buf), launch_index);
}

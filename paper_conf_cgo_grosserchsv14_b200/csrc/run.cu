// run.cu -- the host driver (a7): stencil_run.
//
// "The T dimension is mapped to the host code, where it takes the form of a for loop
// repeatedly iterating over two CUDA kernels -- one kernel for p = 0 and the other one for
// p = 1" (Sec. 4.1).  Each launch-table entry becomes one kernel launch
// on the caller's stream; the grid is the S0 range of that (T, p).
#include <cstring>

#include <cuda_runtime.h>
#include <cstdlib>

#include "internal.h"
#include "kernels/launch.h"

namespace hexs {

static stencil_status cuda_fail(cudaError_t e, const char* where) {
  return fail(STENCIL_E_CUDA, std::string(where) + ": " + cudaGetErrorString(e));
}

#define HEXS_CUDA(call, where)                    \
  do {                                            \
    cudaError_t e_ = (call);                      \
    if (e_ != cudaSuccess) return cuda_fail(e_, where); \
  } while (0)

// K_LINEAR terms: element offsets of the access set in the descriptor's order
static void fill_linear(const Desc& d, LinearTerms& L) {
  L = LinearTerms{};
  if (d.kind != STENCIL_LINEAR) return;
  L.n = (int)d.lcoef.size();
  L.R = d.radius;
  int64_t st[3] = {1, 1, 1};
  st[d.dims - 1] = 1;
  for (int q = d.dims - 2; q >= 0; --q) st[q] = st[q + 1] * d.ext[q + 1];
  for (int k = 0; k < L.n; ++k) {
    int64_t delta = 0;
    for (int q = 0; q < d.dims; ++q) delta += (int64_t)d.loff[k * d.dims + q] * st[q];
    L.delta[k] = delta;
    L.coef[k] = d.lcoef[k];
  }
}

static void fill_generic(const Plan& p, const Launch& l, GenericArgs& g) {
  const Desc& d = p.desc;
  g.dims = d.dims;
  g.hd = p.hd;
  g.ncls = p.ncls;
  for (int q = 0; q < 3; ++q) g.N[q] = q < d.dims ? d.ext[q] : 1;
  g.st[d.dims - 1] = 1;
  for (int q = d.dims - 2; q >= 0; --q) g.st[q] = g.st[q + 1] * d.ext[q + 1];
  for (int q = 0; q < 2; ++q) {
    g.cls[q] = p.cls[q];
    g.dcls[q] = p.dcls[q];
    g.w[q] = p.w[q];
    g.Slo[q] = l.Slo[q];
    g.Shi[q] = l.Shi[q];
  }
  g.tau0 = l.tau0;
  g.a_lo = l.a_lo;
  g.a_hi = l.a_hi;
  g.S0_lo = l.S0_lo;
  g.row_off = l.row_off;
  g.W = p.W;
  g.k0 = d.coef[0];
  g.k1 = d.coef[1];
  for (int a = 0; a < p.H; ++a) {
    g.lo[a] = p.lo[a];
    g.hi[a] = p.hi[a];
  }
  fill_linear(d, g.lin);
}

Plan::~Plan() {
  if (dist) dist_free(dist);
  for (void* e : prof_events)
    if (e) cudaEventDestroy(static_cast<cudaEvent_t>(e));
  for (auto& gr : graphs)
    if (gr.exec) cudaGraphExecDestroy(static_cast<cudaGraphExec_t>(gr.exec));
  if (capture_stream) cudaStreamDestroy(static_cast<cudaStream_t>(capture_stream));
}

static int64_t launches_per_run(const Plan& p) {
  return p.executor == EXEC_NAIVE ? p.tau_levels : (int64_t)p.launches.size();
}

stencil_status run_plan(Plan& p, const void* const* in, void* const* out, void* stream_) {
  const Desc& d = p.desc;
  // optional kernel-region events (stencil_plan_profile): one event before the first phase
  // kernel of the run and one after the last, on the run's stream
  cudaEvent_t* ev = nullptr;
  if (p.prof_runs > 0 && p.prof_used < p.prof_runs) {
    ev = reinterpret_cast<cudaEvent_t*>(p.prof_events.data()) + (size_t)p.prof_used * 2;
    p.prof_used++;
  }
  const int64_t n_launch = launches_per_run(p);
  int64_t li = 0;
  auto ev_begin = [&](cudaStream_t st) {
    if (ev && li == 0) cudaEventRecord(ev[0], st);
  };
  auto ev_end = [&](cudaStream_t st) {
    ++li;
    if (ev && li == n_launch) cudaEventRecord(ev[1], st);
  };
  cudaStream_t s = static_cast<cudaStream_t>(stream_);
  const size_t bytes = (size_t)d.points() * d.elem();
  // HEXS_F3_CHAIN=0: 3D launches strictly one after the other (no cross-launch overlap)
  static const bool f3_chain = [] {
    const char* e = getenv("HEXS_F3_CHAIN");
    return !(e && e[0] == '0');
  }();
  int dev = -1;
  HEXS_CUDA(cudaGetDevice(&dev), "stencil_run: no CUDA device");
  HEXS_CUDA(cudaGetLastError(), "stencil_run: pending CUDA error");

  for (int f = 0; f < d.nfields; ++f) {
    if (!in[f] || !out[f]) return fail(STENCIL_E_INVALID, "stencil_run: NULL field pointer");
    if ((reinterpret_cast<uintptr_t>(in[f]) | reinterpret_cast<uintptr_t>(out[f])) % 16)
      return fail(STENCIL_E_INVALID, "stencil_run: field pointers must be 16-B aligned");
    if (in[f] != out[f])
      HEXS_CUDA(cudaMemcpyAsync(out[f], in[f], bytes, cudaMemcpyDeviceToDevice, s), "stencil_run: copy in->out");
  }
  if (p.T_steps == 0) return STENCIL_OK;

  void* buf[2] = {out[0], p.ws};
  if (d.pingpong) {
    if (!p.ws || p.ws_size < p.ws_bytes)
      return fail(STENCIL_E_INVALID, "stencil_run: workspace not set (stencil_plan_set_workspace)");
    // both ping-pong buffers start as `in`, so Dirichlet cells are valid in either parity
    HEXS_CUDA(cudaMemcpyAsync(p.ws, out[0], bytes, cudaMemcpyDeviceToDevice, s), "stencil_run: init workspace");
  }

  if (p.executor == EXEC_NAIVE) {
    NaiveArgs a{};
    for (int q = 0; q < 3; ++q) a.N[q] = q < d.dims ? d.ext[q] : 1;
    a.k0 = d.coef[0];
    a.k1 = d.coef[1];
    fill_linear(d, a.lin);
    for (int f = 0; f < d.nfields; ++f) a.f[f] = out[f];
    for (int64_t tau = 0; tau < p.tau_levels; ++tau) {
      a.src = buf[tau & 1];
      a.dst = buf[(tau + 1) & 1];
      a.stmt = (int)(tau % (int64_t)d.stmts.size());
      ev_begin(s);
      HEXS_CUDA(launch_naive(d.kind, d.dtype, d.dims, a, s), "stencil_run: naive kernel launch");
      ev_end(s);
    }
  } else {
    if (p.wavefront)
      HEXS_CUDA(cudaMemsetAsync(static_cast<char*>(p.ws) + p.flag_off, 0, p.flag_bytes, s),
                "stencil_run: reset tile flags");
    if (p.executor == EXEC_STREAM3D)
      HEXS_CUDA(cudaMemsetAsync(static_cast<char*>(p.ws) + p.s3_ctr_off, 0, p.s3_ctr_bytes, s),
                "stencil_run: reset strip progress counters");
    int64_t launch_k = 0;
    for (const Launch& l : p.launches) {
      if (p.pre_launch) {  // (k = 0 too: the slab mode's fused exchange seeds the mirrors)
        void* const bufs[2] = {buf[0], buf[1]};
        const stencil_status hs = p.pre_launch(p.pre_launch_ctx, launch_k, bufs, s);
        if (hs != STENCIL_OK) return hs;
      }
      ++launch_k;
      const int a_final = (l.tau0 + l.a_hi + 1 == p.tau_levels) ? l.a_hi : -1;
      const int64_t grid64 = l.S0_hi - l.S0_lo + 1;
      if (grid64 > INT32_MAX) return fail(STENCIL_E_UNSUPPORTED, "stencil_run: grid too large");
      const int grid = (int)grid64;
      ev_begin(s);
      if (p.executor == EXEC_FAST2D) {
        Fast2DArgs a{};
        a.buf[0] = buf[0];
        a.buf[1] = buf[1];
        a.N0 = d.ext[0];
        a.N1 = d.ext[1];
        a.tau0 = l.tau0;
        a.a_lo = l.a_lo;
        a.a_hi = l.a_hi;
        a.a_final = a_final;
        a.S0_lo = l.S0_lo;
        a.row_off = l.row_off;
        a.W = p.W;
        a.k0 = d.coef[0];
        a.k1 = d.coef[1];
        HEXS_CUDA(launch_fast2d(p.variant, a, grid, s), "stencil_run: fast2d kernel launch");
      } else if (p.executor == EXEC_FDTD) {
        FdtdArgs a{};
        for (int f = 0; f < 3; ++f) a.f[f] = out[f];
        a.N0 = d.ext[0];
        a.N1 = d.ext[1];
        a.tau0 = l.tau0;
        a.a_lo = l.a_lo;
        a.a_hi = l.a_hi;
        a.a_final = a_final;
        a.S0_lo = l.S0_lo;
        a.row_off = l.row_off;
        a.W = p.W;
        a.k0 = d.coef[0];
        a.k1 = d.coef[1];
        for (int q = 0; q < p.H; ++q) {
          a.lo[q] = p.lo[q];
          a.hi[q] = p.hi[q];
        }
        HEXS_CUDA(launch_fdtd(p.variant, a, grid, s), "stencil_run: fdtd kernel launch");
      } else if (p.executor == EXEC_STREAM3D) {
        Stream3DArgs a{};
        a.buf[0] = buf[0];
        a.buf[1] = buf[1];
        a.N0 = d.ext[0];
        a.N1 = d.ext[1];
        a.N2 = d.ext[2];
        a.tau0 = l.tau0;
        a.a_lo = l.a_lo;
        a.a_hi = l.a_hi;
        a.a_final = a_final;
        a.S0_lo = l.S0_lo;
        a.row_off = l.row_off;
        a.W = p.W;
        a.L = p.H;
        a.RN = 2 * p.h + p.w0 + 1;
        a.n_str = p.s3_nstr;
        a.n_items = (int)((l.S0_hi - l.S0_lo + 1) * p.s3_nstr);
        a.k0 = d.coef[0];
        a.k1 = d.coef[1];
        char* ws = static_cast<char*>(p.ws);
        a.progress = reinterpret_cast<int*>(ws + p.s3_ctr_off) + l.s3_ctr_first;
        a.ticket = reinterpret_cast<unsigned int*>(a.progress + a.n_items);
        a.scratch = reinterpret_cast<float*>(ws + p.s3_scratch_off);
        HEXS_CUDA(launch_stream3d(p.variant, a, s), "stencil_run: stream3d kernel launch");
      } else if (p.executor == EXEC_ABLATION) {
        AblArgs a{};
        a.buf[0] = buf[0];
        a.buf[1] = buf[1];
        a.N0 = d.ext[0];
        a.N1 = d.ext[1];
        a.N2 = d.ext[2];
        a.tau0 = l.tau0;
        a.a_lo = l.a_lo;
        a.a_hi = l.a_hi;
        a.S0_lo = l.S0_lo;
        a.S0_hi = l.S0_hi;
        a.row_off = l.row_off;
        a.W = p.W;
        a.S1_lo = l.Slo[0];
        a.S2_lo = l.Slo[1];
        a.n1 = (int)(l.Shi[0] - l.Slo[0] + 1);
        a.n2 = (int)(l.Shi[1] - l.Slo[1] + 1);
        a.ctrans1 = p.ctrans[0];
        a.ctrans2 = p.ctrans[1];
        a.YB = p.H + 11;
        a.XB = p.H + 33;
        a.XP = p.variant == ABL_E ? 64 : a.XB;
        a.k0 = d.coef[0];
        a.k1 = d.coef[1];
        for (int q = 0; q < p.H; ++q) {
          a.lo[q] = p.lo[q];
          a.hi[q] = p.hi[q];
        }
        char* ws = static_cast<char*>(p.ws);
        a.progress = reinterpret_cast<int*>(ws + p.flag_off) + l.flag_first;
        a.counter = reinterpret_cast<unsigned int*>(reinterpret_cast<unsigned long long*>(ws + p.counter_off) +
                                                    l.counter_idx);
        HEXS_CUDA(launch_ablation(p.variant, d.kind, a, s), "stencil_run: Table 4 kernel launch");
      } else if (p.executor == EXEC_FAST3D) {
        Fast3DArgs a{};
        a.buf[0] = buf[0];
        a.buf[1] = buf[1];
        a.N0 = d.ext[0];
        a.N1 = d.ext[1];
        a.N2 = d.ext[2];
        a.tau0 = l.tau0;
        a.a_lo = l.a_lo;
        a.a_hi = l.a_hi;
        a.a_final = a_final;
        a.S0_lo = l.S0_lo;
        a.S0_hi = l.S0_hi;
        a.row_off = l.row_off;
        a.W = p.W;
        a.H = p.h;
        a.L = p.H;
        a.Q = p.w0 + 2 * p.h + 3;
        a.S1_lo = l.Slo[0];
        a.n1 = l.Shi[0] - l.Slo[0] + 1;
        a.S2_lo = l.Slo[1];
        a.n2 = l.Shi[1] - l.Slo[1] + 1;
        a.k0 = d.coef[0];
        a.k1 = d.coef[1];
        for (int q = 0; q < p.H; ++q) {
          a.lo[q] = p.lo[q];
          a.hi[q] = p.hi[q];
        }
        char* ws = static_cast<char*>(p.ws);
        a.flags = reinterpret_cast<int*>(ws + p.flag_off) + l.flag_first;
        for (int q = 0; q < 2; ++q) {
          a.mir[q] = p.mir[q];
          a.mir_y0[q] = p.mir_y0[q];
        }
        a.mir_G = p.mir_G;
        a.mir_fence = p.mir_fence;
        a.counter = reinterpret_cast<unsigned long long*>(ws + p.counter_off) + l.counter_idx;
        // chained launches (single GPU): launch k may start while k-1 drains; its tiles acquire
        // the flags of the tiles of k-1 and k-2 they read from (hex3d.cu wait_prev)
        const bool chain = f3_chain && !p.pre_launch && !p.mir[0] && !p.mir[1];
        if (chain) {
          const int64_t k = &l - p.launches.data();
          for (int q = 0; q < 2; ++q) {
            if (k - 1 - q < 0) continue;
            const Launch& pl = p.launches[(size_t)(k - 1 - q)];
            Fast3DPrev& pv = a.prev[q];
            pv.flags = reinterpret_cast<const int*>(ws + p.flag_off) + pl.flag_first;
            pv.done = reinterpret_cast<const unsigned long long*>(ws + p.counter_off) + p.n_counters + pl.counter_idx;
            pv.tau0 = pl.tau0;
            pv.S0_lo = pl.S0_lo;
            pv.S0_hi = pl.S0_hi;
            pv.row_off = pl.row_off;
            pv.S1_lo = pl.Slo[0];
            pv.n1 = pl.Shi[0] - pl.Slo[0] + 1;
            pv.S2_lo = pl.Slo[1];
            pv.n2 = pl.Shi[1] - pl.Slo[1] + 1;
          }
          a.pdl = 1;
          a.done = reinterpret_cast<unsigned long long*>(ws + p.counter_off) + p.n_counters + l.counter_idx;
        }
        HEXS_CUDA(launch_fast3d(p.variant, a, grid, s), "stencil_run: fast3d kernel launch");
      } else {
        GenericArgs g{};
        if (d.pingpong) {
          g.f[0] = buf[0];
          g.f[1] = buf[1];
        } else {
          for (int f = 0; f < 3; ++f) g.f[f] = out[f];
        }
        fill_generic(p, l, g);
        g.S0_hi = l.S0_hi;
        if (p.wavefront) {
          char* ws = static_cast<char*>(p.ws);
          g.wf = 1;
          g.flags = reinterpret_cast<int*>(ws + p.flag_off) + l.flag_first;
          g.counter = reinterpret_cast<unsigned long long*>(ws + p.counter_off) + l.counter_idx;
        }
        HEXS_CUDA(launch_generic(d.kind, d.dtype, g, grid, s), "stencil_run: generic kernel launch");
      }
      ev_end(s);
    }
  }
  // level T_steps lives in buffer T_steps % 2
  if (d.pingpong && (p.tau_levels & 1))
    HEXS_CUDA(cudaMemcpyAsync(out[0], p.ws, bytes, cudaMemcpyDeviceToDevice, s), "stencil_run: copy result");
  return STENCIL_OK;
}

}  // namespace hexs

using namespace hexs;

extern "C" stencil_status stencil_run(stencil_plan_t plan, const void* const* in, void* const* out,
                                      int64_t T_steps, void* stream) {
  clear_error();
  Plan* p = reinterpret_cast<Plan*>(plan);
  if (!p || p->magic != kPlanMagic) return fail(STENCIL_E_INVALID, "stencil_run: bad plan");
  if (!in || !out) return fail(STENCIL_E_INVALID, "stencil_run: in/out is NULL");
  if (T_steps != p->T_steps) return fail(STENCIL_E_INVALID, "stencil_run: T_steps differs from the plan's");
  if (p->dist) return run_dist(*p, in, out, stream);  // multi-GPU slab mode (dist.cpp)
  // Replay a captured CUDA graph of the whole run when the pointers match an earlier run (and no
  // profiling is requested); the first run is eager (kernel attributes, occupancy queries), the
  // second is captured on a private stream and replayed from then on.  HEXS_NO_GRAPH=1 disables.
  static const bool no_graph = std::getenv("HEXS_NO_GRAPH") && std::atoi(std::getenv("HEXS_NO_GRAPH")) != 0;
  if (no_graph || p->prof_runs > 0 || p->T_steps == 0) return run_plan(*p, in, out, stream);
  std::vector<const void*> key;
  for (int f = 0; f < p->desc.nfields; ++f) {
    if (!in[f] || !out[f]) return fail(STENCIL_E_INVALID, "stencil_run: NULL field pointer");
    key.push_back(in[f]);
    key.push_back(out[f]);
  }
  key.push_back(p->ws);
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  for (auto& gr : p->graphs)
    if (gr.key == key) {
      HEXS_CUDA(cudaGraphLaunch(static_cast<cudaGraphExec_t>(gr.exec), s), "stencil_run: graph launch");
      return STENCIL_OK;
    }
  if (p->eager_runs++ == 0 || p->graphs.size() >= 8) return run_plan(*p, in, out, stream);
  // the private capture stream lives on the device the plan currently runs on
  int dev = -1;
  HEXS_CUDA(cudaGetDevice(&dev), "stencil_run: no CUDA device");
  if (p->capture_stream && p->capture_dev != dev) {
    cudaStreamDestroy(static_cast<cudaStream_t>(p->capture_stream));
    p->capture_stream = nullptr;
  }
  if (!p->capture_stream) {
    cudaStream_t cs = nullptr;
    HEXS_CUDA(cudaStreamCreateWithFlags(&cs, cudaStreamNonBlocking), "stencil_run: capture stream");
    p->capture_stream = cs;
    p->capture_dev = dev;
  }
  cudaStream_t cs = static_cast<cudaStream_t>(p->capture_stream);
  HEXS_CUDA(cudaStreamBeginCapture(cs, cudaStreamCaptureModeThreadLocal), "stencil_run: begin capture");
  const stencil_status st = run_plan(*p, in, out, cs);
  cudaGraph_t graph = nullptr;
  const cudaError_t ec = cudaStreamEndCapture(cs, &graph);
  if (st != STENCIL_OK) {
    // a launch failed while capturing: drop the partial graph and run eagerly on the
    // caller's stream (a genuine error surfaces again there)
    if (graph) cudaGraphDestroy(graph);
    cudaGetLastError();
    clear_error();
    return run_plan(*p, in, out, stream);
  }
  if (ec != cudaSuccess || !graph) {
    cudaGetLastError();
    return run_plan(*p, in, out, stream);  // capture unsupported here: stay eager
  }
  cudaGraphExec_t exec = nullptr;
  const cudaError_t ei = cudaGraphInstantiate(&exec, graph, 0);
  cudaGraphDestroy(graph);
  if (ei != cudaSuccess) {
    cudaGetLastError();
    return run_plan(*p, in, out, stream);
  }
  p->graphs.push_back({key, exec});
  HEXS_CUDA(cudaGraphLaunch(exec, s), "stencil_run: graph launch");
  return STENCIL_OK;
}

extern "C" stencil_status stencil_plan_profile(stencil_plan_t plan, int max_runs) {
  clear_error();
  Plan* p = reinterpret_cast<Plan*>(plan);
  if (!p || p->magic != kPlanMagic || max_runs < 0) return fail(STENCIL_E_INVALID, "stencil_plan_profile: bad arguments");
  for (void* e : p->prof_events)
    if (e) cudaEventDestroy(static_cast<cudaEvent_t>(e));
  p->prof_events.clear();
  p->prof_runs = 0;
  p->prof_used = 0;
  if (max_runs == 0) return STENCIL_OK;
  const size_t n = (size_t)max_runs * 2;
  p->prof_events.assign(n, nullptr);
  for (size_t i = 0; i < n; ++i) {
    cudaEvent_t e;
    cudaError_t r = cudaEventCreate(&e);
    if (r != cudaSuccess) return cuda_fail(r, "stencil_plan_profile: cudaEventCreate");
    p->prof_events[i] = e;
  }
  p->prof_runs = max_runs;
  return STENCIL_OK;
}

extern "C" stencil_status stencil_plan_profile_read(stencil_plan_t plan, double* kernel_ms, int64_t* launches,
                                                    double* max_launch_ms) {
  clear_error();
  Plan* p = reinterpret_cast<Plan*>(plan);
  if (!p || p->magic != kPlanMagic || !kernel_ms || !launches || !max_launch_ms)
    return fail(STENCIL_E_INVALID, "stencil_plan_profile_read: bad arguments");
  const int64_t runs = p->prof_used, per = launches_per_run(*p);
  double total = 0, mx = 0;
  cudaEvent_t* ev = reinterpret_cast<cudaEvent_t*>(p->prof_events.data());
  for (int64_t i = 0; i < runs && per > 0; ++i) {
    HEXS_CUDA(cudaEventSynchronize(ev[2 * i + 1]), "stencil_plan_profile_read: sync");
    float ms = 0;
    HEXS_CUDA(cudaEventElapsedTime(&ms, ev[2 * i], ev[2 * i + 1]), "stencil_plan_profile_read: elapsed");
    total += ms;
    if (ms > mx) mx = ms;
  }
  *kernel_ms = total;
  *launches = per > 0 ? runs * per : 0;
  *max_launch_ms = mx;
  p->prof_used = 0;
  return STENCIL_OK;
}

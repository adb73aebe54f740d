// internal.h -- library-internal data structures of libhexstencil (host side).
#pragma once
#include <cstddef>
#include <cstdint>
#include <string>
#include <vector>

#include "../../include/stencil.h"

namespace hexs {

constexpr uint32_t kDescMagic = 0x48584453u;  // "HXDS"
constexpr uint32_t kPlanMagic = 0x48585053u;  // "HXPS"
constexpr int kMaxLevels = 64;                // max 2h+2 supported by the kernels
constexpr int kStream3DNXPlan = 64;           // = kernels/launch.h kStream3DNX (strip width)
constexpr int kStream3DRSPlan = 32;           // = kernels/launch.h kStream3DRS (carry ring depth)

// A rational number n/d, d > 0, reduced.
struct Rat {
  int64_t n = 0, d = 1;
};
Rat make_rat(int64_t n, int64_t d);
bool rat_less(const Rat& a, const Rat& b);
int64_t floor_div(int64_t a, int64_t b);
int64_t ceil_div(int64_t a, int64_t b);

// The statement model of Sec. 3.2: an outer time loop around k >= 1
// perfect nests; statement i writes field `write` at offset 0 and reads `reads`.
struct Access {
  int field;
  int off[3];
};
struct Stmt {
  int write;
  std::vector<Access> reads;
  int lo[3];  // domain per dim: [lo, N + hi)
  int hi[3];
};

struct Desc {
  uint32_t magic = kDescMagic;
  int dims = 0;
  int64_t ext[3] = {1, 1, 1};
  int kind = 0;
  int radius = 1;
  int dtype = 0;
  double coef[4] = {0, 0, 0, 0};
  int ncoef = 0;
  int nfields = 1;
  bool pingpong = true;
  std::vector<Stmt> stmts;
  // STENCIL_LINEAR: the access set (n x dims offsets, slow -> fast) and its coefficients
  std::vector<int> loff;
  std::vector<double> lcoef;
  size_t elem() const { return dtype == STENCIL_F64 ? 8 : 4; }
  int64_t points() const { return ext[0] * ext[1] * (dims == 3 ? ext[2] : 1); }
};

// Distance vectors (dtau, ds...) of the canonical schedule (dependence analysis, a1).
std::vector<std::vector<int64_t>> dependence_distances(const Desc& d);

struct Launch {
  int64_t T;
  int phase;
  int a_lo, a_hi;
  int64_t tau0;
  int64_t S0_lo, S0_hi;
  int64_t row_off;
  // classical tile index ranges (generic executor)
  int64_t Slo[2], Shi[2];
  // wavefront executors: first tile flag and work counter of this launch in the workspace
  int64_t flag_first = 0, counter_idx = 0;
  // stream3d: first progress counter of this launch (its ticket follows the launch's counters)
  int64_t s3_ctr_first = 0;
};

enum Executor { EXEC_GENERIC = 1, EXEC_NAIVE = 2, EXEC_FAST2D = 3, EXEC_FDTD = 4, EXEC_FAST3D = 5, EXEC_STREAM3D = 6,
               EXEC_ABLATION = 7 };

// Multi-GPU slab mode (dist.cpp): partition, time blocks, local block plans, NCCL state.
struct DistLayout {
  int rank, nranks, part_dim, h;
  int64_t own_lo, own_hi, loc_lo, loc_hi, ghost, time_block, n_blocks;
  double ghost_fraction;
};
struct DistState;
void dist_free(DistState* d);

struct Plan {
  uint32_t magic = kPlanMagic;
  DistState* dist = nullptr;  // non-null: a stencil_plan_dist plan (stencil_run runs the slab mode)
  Desc desc;
  int64_t T_steps = 0, tau_levels = 0;
  int hd = 0;           // hexagonal dimension
  int ncls = 0;         // number of classical dims
  int cls[2] = {0, 0};  // classical dims (slow -> fast)
  Rat d0, d1;           // cone slopes along hd
  int dcls[2] = {0, 0}; // integer classical skews delta1_i
  int ctrans[2] = {0, 0};  // classical tile translation offsets (Sec. 4.2.3)
  int h = 0, w0 = 0, w[2] = {1, 1};
  int H = 0, W = 0, F0 = 0, F1 = 0, c = 0;
  int64_t hex_origin = 0;  // global coordinate of local row 0 along hd (slab plans)
  // called before every phase-kernel launch k >= 1 with the two ping-pong buffers (multi-GPU
  // slab mode: the per-launch ghost exchange); nullptr = none
  stencil_status (*pre_launch)(void* ctx, int64_t k, void* const* bufs, void* stream) = nullptr;
  void* pre_launch_ctx = nullptr;
  // fused halo stores of the 3D tile-wavefront kernel (slab mode, set per run by dist.cpp):
  // neighbour s's mirror base, the first local line of the zone it mirrors, the zone width
  void* mir[2] = {nullptr, nullptr};
  int mir_y0[2] = {0, 0};
  int mir_G = 0;
  int mir_fence = 1;
  std::vector<int32_t> lo, hi;  // hexagon rows per level a
  std::vector<Launch> launches;
  int executor = EXEC_GENERIC;
  int variant = 0;  // fast-kernel instantiation id
  int64_t tile_points = 0, tile_in = 0, tile_out = 0;
  bool wavefront = false;      // generic executor: classical tiles as a dependence wavefront
  size_t flag_off = 0, counter_off = 0, flag_bytes = 0;  // workspace layout (wavefront)
  int64_t n_counters = 0;  // ticket counters; the completed-tile counters follow them
  // stream3d: per-launch progress counters + ticket (zeroed per run), carry scratch
  size_t s3_ctr_off = 0, s3_ctr_bytes = 0, s3_scratch_off = 0;
  int s3_nstr = 0;
  size_t ws_bytes = 0;
  void* ws = nullptr;
  size_t ws_size = 0;
  // profiling: event pairs around each launch for up to prof_runs runs
  int prof_runs = 0, prof_used = 0;
  std::vector<void*> prof_events;  // cudaEvent_t, 2 per launch per run
  // CUDA graphs of whole runs (the launch sequence is fixed by the plan): keyed by the field,
  // workspace pointers; replayed on the caller's stream (a run is launch-bound on small grids)
  struct GraphEntry {
    std::vector<const void*> key;
    void* exec = nullptr;  // cudaGraphExec_t
  };
  std::vector<GraphEntry> graphs;
  int eager_runs = 0;      // runs executed eagerly (the first one sets kernel attributes)
  void* capture_stream = nullptr;
  int capture_dev = -1;  // device the capture stream was created on
  ~Plan();
};

// Error reporting (thread-local message).
stencil_status fail(stencil_status s, const std::string& msg);
void clear_error();

// plan.cpp
// hex_origin: the global coordinate of local row 0 along the hexagonal dimension -- a local plan
// of a slab (multi-GPU) keeps the global hexagon tiling (Sec. 4.2.3's tile translation offset)
stencil_status build_plan(const Desc& d, int64_t T_steps, const stencil_tile_t* tile, Plan** out,
                          int64_t hex_origin = 0);
bool schedule_of(const Plan& p, int64_t tau, const int64_t* s, int64_t* sched);

// run.cu
stencil_status run_plan(Plan& p, const void* const* in, void* const* out, void* stream);
// dist.cpp
stencil_status run_dist(Plan& p, const void* const* in, void* const* out, void* stream);
stencil_status dist_set_workspace(Plan& p, void* dev_ptr, size_t bytes);
void dist_fill_info(const Plan& p, stencil_plan_info_t& o);

// Fast-kernel registry (kernels/*.cu): returns variant id >= 0 or -1 if not instantiated.
int fast2d_variant(int kind, int dtype, int h, int w0, int w1);
int fast2d_chunk_width(int variant);  // classical tile width w1 the kernel streams
int fdtd_variant(int dtype, int h, int w0);
int fdtd_ctas_per_sm();
int fast3d_variant(int kind, int dtype, int h, int w0, int wy);
int fast3d_tile(int variant, int* wy, int* wx);
bool fast3d_variant_matches(int variant, int kind, int dtype, int h, int w0);
int stream3d_variant(int kind, int dtype, int h, int w0);
int fast2d_variant_count();
bool fast2d_variant_info(int variant, int* kind, int* dtype, int* h, int* w0);
int fast3d_variant_count();
bool fast3d_variant_info(int variant, int* kind, int* dtype, int* h, int* w0);

// tilemodel.cpp: the tile-size model of Sec. 3.7 (load-to-compute ratio) with the on-chip
// (instruction cache) and CTA-count terms of the B200 kernels
enum TileFamily { FAMILY_GENERIC = 0, FAMILY_FAST2D = 1, FAMILY_FAST3D = 2 };
struct TileEval {
  int h, w0;
  int64_t points, in, out;  // per classical column of one full hexagon
  double bytes_per_update;  // word * (In + Out) / points
  double body_bytes;        // unrolled level bodies of the fast kernels (instruction cache)
  double code_eff;          // min(1, capacity / body)^3
  int64_t ctas, slots;      // CTAs of a full launch and resident slots
  double wave_eff;          // ctas / (waves * slots)
  double rate;              // predicted relative rate (updates / s, up to a constant)
};
bool tile_eval(const Desc& d, int hd, const Rat& d0, const Rat& d1, int h, int w0, int family, TileEval* out);
bool tile_select(const Desc& d, int hd, const Rat& d0, const Rat& d1, int family, int* h, int* w0);
int stream3d_carry_block(int variant);  // floats per (strip, step) carry block

}  // namespace hexs

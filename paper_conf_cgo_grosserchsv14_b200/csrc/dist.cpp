// dist.cpp -- multi-GPU slab mode of the C ABI: one process per GPU,
// one non-innermost grid dimension (3D default: y, a classically tiled dimension) slab-partitioned
// over the ranks, halos exchanged with NCCL send/recv over NVLink once per phase launch (time tile).
//
// The paper's method is single-GPU: its host loop iterates the two phase kernels over the
// whole grid (Sec. 4.1).  Here every rank runs exactly that host loop -- the
// SAME launch table (T, p) as the global run -- over its local slab, and the ranks exchange
// halos between consecutive launches:
//   * rank q owns indices [own_lo, own_hi) of the partitioned dimension (an even split) and
//     stores the local slab [loc_lo, loc_hi) = owned indices plus G = radius * (2h+2) ghost
//     indices on every side that is not a global boundary (the halo width "radius x time-tile
//     depth");
//   * the local plan keeps the GLOBAL hexagon tiling: when the partitioned dimension is the
//     hexagonal one its rows are translated by loc_lo (Sec. 4.2.3's tile translation offset);
//     when it is a classical one (the 3D default, y) the hexagonal dimension is whole on every
//     rank and the launch table is the global one as is -- which levels a launch computes at a
//     point depends only on its (t, hexagonal) coordinates, never on the classical tiling -- so
//     after every launch each point of the slab holds the same level as in a single-GPU run;
//   * before every launch but the first, the ghost indices of BOTH ping-pong buffers are
//     refreshed from the neighbours' owned ones (ncclGroupStart; ncclSend / ncclRecv to rank -1
//     and rank +1; ncclGroupEnd), on a communication stream ordered against the compute stream
//     by events; a partition of dimension > 0 is strided in memory, so its slabs are packed into
//     / unpacked from a staging area of the workspace with 2-D copies on the same stream; the
//     outermost local indices act as fixed (Dirichlet) cells, and a launch spans at most 2h+2
//     levels, so its wrong values never travel further than G indices: every owned point is
//     exact after every launch.  The only redundant work is the ghost slabs (2G / owned of the
//     compute); there are no time-block cuts (the schedule is continuous).
// NCCL is loaded at run time (dlopen of the libnccl.so.2 the process already uses, e.g.
// PyTorch's), so single-GPU use of the library never needs it; PyTorch only broadcasts the
// 128-byte unique id (stencil_dist_unique_id on rank 0).
#include <dlfcn.h>

#include <algorithm>
#include <cstdlib>
#include <cstring>
#include <map>
#include <memory>
#include <mutex>
#include <new>
#include <string>
#include <vector>

#include <cuda_runtime.h>
#include <nccl.h>

#include "internal.h"
#include "kernels/launch.h"

namespace hexs {

namespace {

struct NcclApi {
  void* handle = nullptr;
  ncclResult_t (*GetUniqueId)(ncclUniqueId*) = nullptr;
  ncclResult_t (*CommInitRank)(ncclComm_t*, int, ncclUniqueId, int) = nullptr;
  ncclResult_t (*CommDestroy)(ncclComm_t) = nullptr;
  ncclResult_t (*GroupStart)() = nullptr;
  ncclResult_t (*GroupEnd)() = nullptr;
  ncclResult_t (*Send)(const void*, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
  ncclResult_t (*Recv)(void*, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
  const char* (*GetErrorString)(ncclResult_t) = nullptr;
  ncclResult_t (*CommGetAsyncError)(ncclComm_t, ncclResult_t*) = nullptr;
  // symmetric memory (NCCL >= 2.27): device-initiated halo stores through LSA pointers
  ncclResult_t (*MemAlloc)(void**, size_t) = nullptr;
  ncclResult_t (*MemFree)(void*) = nullptr;
  ncclResult_t (*WindowRegister)(ncclComm_t, void*, size_t, ncclWindow_t*, int) = nullptr;
  ncclResult_t (*WindowDeregister)(ncclComm_t, ncclWindow_t) = nullptr;
  ncclResult_t (*AllReduce)(const void*, void*, size_t, ncclDataType_t, ncclRedOp_t, ncclComm_t, cudaStream_t) = nullptr;
  std::string error;
};

// Load NCCL once: HEXS_NCCL_LIB if set, else the libnccl.so.2 already mapped into the process
// (PyTorch's), else the dynamic linker's.
NcclApi* nccl_api() {
  static NcclApi api;
  static bool tried = false;
  if (tried) return api.handle ? &api : nullptr;
  tried = true;
  const char* env = std::getenv("HEXS_NCCL_LIB");
  void* h = nullptr;
  if (env && *env) h = dlopen(env, RTLD_NOW | RTLD_GLOBAL);
  if (!h) h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_NOLOAD | RTLD_GLOBAL);
  if (!h) h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
  if (!h) h = dlopen("libnccl.so", RTLD_NOW | RTLD_GLOBAL);
  if (!h) {
    const char* e = dlerror();
    api.error = std::string("cannot load libnccl.so.2: ") + (e ? e : "?");
    return nullptr;
  }
  auto sym = [&](const char* name) { return dlsym(h, name); };
  api.GetUniqueId = reinterpret_cast<decltype(api.GetUniqueId)>(sym("ncclGetUniqueId"));
  api.CommInitRank = reinterpret_cast<decltype(api.CommInitRank)>(sym("ncclCommInitRank"));
  api.CommDestroy = reinterpret_cast<decltype(api.CommDestroy)>(sym("ncclCommDestroy"));
  api.GroupStart = reinterpret_cast<decltype(api.GroupStart)>(sym("ncclGroupStart"));
  api.GroupEnd = reinterpret_cast<decltype(api.GroupEnd)>(sym("ncclGroupEnd"));
  api.Send = reinterpret_cast<decltype(api.Send)>(sym("ncclSend"));
  api.Recv = reinterpret_cast<decltype(api.Recv)>(sym("ncclRecv"));
  api.GetErrorString = reinterpret_cast<decltype(api.GetErrorString)>(sym("ncclGetErrorString"));
  api.CommGetAsyncError = reinterpret_cast<decltype(api.CommGetAsyncError)>(sym("ncclCommGetAsyncError"));
  api.MemAlloc = reinterpret_cast<decltype(api.MemAlloc)>(sym("ncclMemAlloc"));
  api.MemFree = reinterpret_cast<decltype(api.MemFree)>(sym("ncclMemFree"));
  api.WindowRegister = reinterpret_cast<decltype(api.WindowRegister)>(sym("ncclCommWindowRegister"));
  api.WindowDeregister = reinterpret_cast<decltype(api.WindowDeregister)>(sym("ncclCommWindowDeregister"));
  api.AllReduce = reinterpret_cast<decltype(api.AllReduce)>(sym("ncclAllReduce"));
  if (!api.GetUniqueId || !api.CommInitRank || !api.CommDestroy || !api.GroupStart || !api.GroupEnd ||
      !api.Send || !api.Recv || !api.GetErrorString) {
    api.error = "libnccl.so.2 lacks a required symbol";
    return nullptr;
  }
  api.handle = h;
  return &api;
}

stencil_status nccl_fail(NcclApi* a, ncclResult_t r, const char* where) {
  return fail(STENCIL_E_NCCL, std::string(where) + ": " + (a && a->GetErrorString ? a->GetErrorString(r) : "NCCL error"));
}

Plan* as_plan(stencil_plan_t h) {
  Plan* p = reinterpret_cast<Plan*>(h);
  return (p && p->magic == kPlanMagic) ? p : nullptr;
}

}  // namespace

struct DistState {
  DistLayout lay;
  std::vector<int64_t> blocks;                     // (one entry: T_steps; kept for the API)
  std::vector<std::pair<int64_t, Plan*>> bplans;   // the local plan (one, T_steps long)
  Desc local;                                      // descriptor of the local slab
  int64_t global_n = 0;                            // global extent of the partitioned dimension
  int64_t n_outer = 1;                             // product of the extents before it
  size_t line_bytes = 0;                           // bytes of one index of it (extents after it)
  size_t local_ws = 0;                             // the local plan's workspace (256-B rounded)
  size_t stage_bytes = 0;                          // halo staging area after it (strided partitions)
  char* stage = nullptr;
  // Needed-state lists (hexagonal dimension 0 whole, a classical dimension partitioned): before
  // launch k, outer index z (the hexagonal coordinate) holds level L(z) in buffer L(z) % 2 and
  // L(z)-1 in the other; the next launch reads the older value only where a z-neighbour is
  // behind (it computes level L(z) from it).  rows[k][b] = the z whose buffer-b halo lines are
  // read; only those travel (~68 % of both buffers for the (3, 7) hexagon).
  std::vector<int> row_table;                      // flat: per launch k >= 1, buffer 0 then 1
  std::vector<std::pair<int64_t, int64_t>> row_span;  // (offset, count) per (k, b)
  size_t rows_off = 0, rows_bytes = 0;             // the table's copy in the workspace
  int* rows_dev = nullptr;
  // Device-initiated exchange (default for nranks > 1 when NCCL symmetric windows work, or in
  // loopback mode HEXS_DIST_LOOPBACK=1: the ranks are plans of one process on one device): each
  // rank owns a receive area [slot k%2][side: from lower, from upper][buffer] x halo bytes + two
  // flags + a block counter; the sender's kernel stores straight into the neighbour's area.
  bool p2p = false, loopback = false;
  // fused: the 3D tile-wavefront kernel itself stores its send-zone lines into the neighbours'
  // mirrors while it computes (the transfer overlaps the launch); the boundary keeps only two
  // flag handshakes and a local scatter
  bool fused = false;
  char* recv = nullptr;
  size_t recv_bytes = 0, recv_halo = 0, flag_off = 0;
  void* win = nullptr;                      // ncclWindow_t of `recv`
  char* peer_recv[2] = {nullptr, nullptr};  // the lower / upper neighbour's receive area
  unsigned int done_count = 0;              // host mirror of the send kernel's block counter
  int64_t runs = 0;                         // completed stencil_runs (flag sequence base)
  std::string group;                        // loopback registry key
  void* comm = nullptr;                            // ncclComm_t
  cudaStream_t comm_stream = nullptr;
  cudaEvent_t ev_ready = nullptr, ev_done = nullptr;
  int comm_dev = -1;
  bool emulate = false;  // HEXS_DIST_EMULATE: a rank's compute alone (no communicator)
  bool emulate_copies = false;  // HEXS_DIST_EMULATE=2: plus the halo copies, a local copy as the wire
  ~DistState();
  void release_p2p();
  void destroy_rest() {
    for (auto& bp : bplans) delete bp.second;
    if (comm) {
      if (NcclApi* a = nccl_api()) a->CommDestroy(static_cast<ncclComm_t>(comm));
    }
    if (ev_ready) cudaEventDestroy(ev_ready);
    if (ev_done) cudaEventDestroy(ev_done);
    if (comm_stream) cudaStreamDestroy(comm_stream);
  }
  Plan* plan_for(int64_t len) const {
    for (auto& bp : bplans)
      if (bp.first == len) return bp.second;
    return nullptr;
  }
};

// loopback registry: the ranks of one group (keyed by the unique id) in this process
static std::mutex g_loop_mu;
static std::map<std::string, std::vector<DistState*>> g_loop;

void DistState::release_p2p() {
  if (loopback && !group.empty()) {
    std::lock_guard<std::mutex> lk(g_loop_mu);
    auto it = g_loop.find(group);
    if (it != g_loop.end()) {
      for (auto& q : it->second)
        if (q == this) q = nullptr;
    }
  }
  if (recv) {
    NcclApi* a = nccl_api();
    if (win && a && a->WindowDeregister) a->WindowDeregister(static_cast<ncclComm_t>(comm), static_cast<ncclWindow_t>(win));
    if (loopback) cudaFree(recv);
    else if (a && a->MemFree) a->MemFree(recv);
  }
  recv = nullptr;
  win = nullptr;
}

DistState::~DistState() {
  release_p2p();
  destroy_rest();
}

void dist_free(DistState* d) { delete d; }

// stencil_plan_info of a distributed plan: the primary block plan's schedule and tile, the
// whole run's steps, launches and this rank's owned updates.
void dist_fill_info(const Plan& p, stencil_plan_info_t& o) {
  const DistState& s = *p.dist;
  int64_t launches = 0;
  for (int64_t len : s.blocks) {
    const Plan* bp = s.plan_for(len);
    launches += bp->executor == EXEC_NAIVE ? bp->tau_levels : (int64_t)bp->launches.size();
  }
  o.n_launches = launches;
  o.T_steps = p.T_steps;
  o.tau_levels = p.tau_levels;
  const int pd = s.lay.part_dim, r = s.local.radius;
  int64_t interior = 1;
  for (int q = 0; q < s.local.dims; ++q)
    if (q != pd) interior *= s.local.ext[q] - 2 * r;
  const int64_t glo = std::max<int64_t>(s.lay.own_lo, r);
  const int64_t ghi = std::min<int64_t>(s.lay.own_hi, s.global_n - r);  // global edge cells are Dirichlet
  o.updates = std::max<int64_t>(0, ghi - glo) * interior * p.T_steps;
  o.workspace_bytes = p.ws_bytes;
}

// The tile of the local plans: the caller's, else the class default the planner picks for the
// GLOBAL grid (heat-3D 1024^3: (3, 7) -- measured per rank with y slabs it beats the shallower
// (2, 7) at every rank count despite its larger ghost share, 12.5 % vs 9.4 % at 128 lines/rank:
// DESIGN.md §7).  Always returned explicit (h, w0), so every rank's local plan and the layout
// share one hexagon (one tiling).
stencil_tile_t dist_local_tile(const Desc& d, const stencil_tile_t* tile, int nranks) {
  (void)nranks;
  stencil_tile_t lt{};
  lt.hex_dim = -1;
  if (tile) lt = *tile;
  if (lt.h || lt.w0) return lt;  // an explicit hexagon
  Plan* probe = nullptr;
  if (build_plan(d, 1, &lt, &probe) == STENCIL_OK) {
    lt.h = probe->h;
    lt.w0 = probe->w0;
    if (lt.hex_dim < 0) lt.hex_dim = probe->hd;
    delete probe;
  }
  return lt;
}

// The needed-state row lists of a local plan whose hexagonal dimension 0 is whole (a classical
// dimension part_dim > 0 partitioned): before launch k >= 1, z holds level L(z) in buffer
// L(z) % 2 and L(z) - 1 in the other; launch k reads the older value only where a z-neighbour is
// behind (it computes level L(z) from it -- adjacent levels differ by at most one, or the
// ping-pong WAR order would be broken).  table: per k >= 1, the z of buffer 0, then buffer 1;
// span[2 (k-1) + b] = (offset, count).  false if the rule does not apply.
bool halo_rows_table(const Plan& lp, int part_dim, std::vector<int>& table,
                     std::vector<std::pair<int64_t, int64_t>>& span) {
  table.clear();
  span.clear();
  if (lp.hd != 0 || part_dim <= 0 || lp.executor == EXEC_NAIVE || lp.desc.nfields != 1 || lp.desc.dims < 2)
    return false;
  const int64_t Z = lp.desc.ext[0];
  std::vector<int64_t> lev(Z, 0);  // level each z holds after the launches so far
  for (size_t k = 0; k < lp.launches.size(); ++k) {
    const Launch& ln = lp.launches[k];
    if (k > 0) {
      for (int b = 0; b < 2; ++b) {
        const int64_t off = (int64_t)table.size();
        for (int64_t z = 0; z < Z; ++z) {
          const bool behind = (z > 0 && lev[z - 1] < lev[z]) || (z + 1 < Z && lev[z + 1] < lev[z]);
          if ((lev[z] & 1) == b || behind) table.push_back((int)z);
        }
        span.push_back({off, (int64_t)table.size() - off});
      }
    }
    for (int a = ln.a_lo; a <= ln.a_hi; ++a)
      for (int64_t S0 = ln.S0_lo; S0 <= ln.S0_hi; ++S0) {
        const int64_t i0 = S0 * lp.W - ln.row_off;
        const int64_t r0 = std::max<int64_t>(i0 + lp.lo[a], 1), r1 = std::min<int64_t>(i0 + lp.hi[a], Z - 2);
        for (int64_t z = r0; z <= r1; ++z) lev[z] = ln.tau0 + a + 1;
      }
  }
  return true;
}

// The slab layout of one rank (host only; shared by stencil_dist_layout and stencil_plan_dist).
stencil_status dist_layout(const Desc& d, int64_t T_steps, const stencil_tile_t* tile, int rank, int nranks,
                           int part_dim, DistLayout* out) {
  if (nranks < 1 || rank < 0 || rank >= nranks) return fail(STENCIL_E_INVALID, "stencil_plan_dist: bad rank / nranks");
  if (part_dim < 0) part_dim = d.dims == 3 ? 1 : 0;  // default: y in 3D (classical), rows in 2D
  if (part_dim > d.dims - 2)
    return fail(STENCIL_E_UNSUPPORTED, "stencil_plan_dist: the partitioned dimension must not be the innermost one");
  if (d.kind == STENCIL_FDTD2D)
    return fail(STENCIL_E_UNSUPPORTED, "stencil_plan_dist: FDTD-2D (three in-place fields) has no slab mode");
  if (T_steps < 0) return fail(STENCIL_E_INVALID, "stencil_plan_dist: T_steps < 0");
  DistLayout L{};
  L.rank = rank;
  L.nranks = nranks;
  L.part_dim = part_dim;
  const int64_t N0 = d.ext[part_dim];
  const int64_t base = N0 / nranks, extra = N0 % nranks;
  L.own_lo = rank * base + std::min<int64_t>(rank, extra);
  L.own_hi = L.own_lo + base + (rank < extra ? 1 : 0);
  const stencil_tile_t lt = dist_local_tile(d, tile, nranks);
  const int h = lt.h;
  const int64_t owned = L.own_hi - L.own_lo;
  // one exchange per phase launch: a launch spans at most 2h+2 levels (one time tile)
  const int64_t D = 2 * (int64_t)h + 2;
  L.time_block = D;
  L.ghost = (int64_t)d.radius * D;
  if (nranks > 1 && owned < L.ghost)
    return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan_dist: a slab is thinner than the ghost width radius*(2h+2)");
  if (nranks > 1 && d.dims == 3 && part_dim == 1 && d.ext[0] < 3)
    return fail(STENCIL_E_INVALID, "stencil_plan_dist: degenerate grid");
  L.loc_lo = std::max<int64_t>(0, L.own_lo - L.ghost);
  L.loc_hi = std::min<int64_t>(N0, L.own_hi + L.ghost);
  L.n_blocks = 0;  // filled by stencil_plan_dist: launches (one exchange before each but the first)
  L.h = h;
  L.ghost_fraction = owned > 0 ? (double)((L.loc_hi - L.loc_lo) - owned) / (double)owned : 0.0;
  *out = L;
  return STENCIL_OK;
}

stencil_status dist_set_workspace(Plan& p, void* dev_ptr, size_t bytes) {
  DistState& s = *p.dist;
  if (bytes < s.local_ws + s.stage_bytes + s.rows_bytes)
    return fail(STENCIL_E_OOM, "stencil_plan_set_workspace: workspace too small");
  for (auto& bp : s.bplans) {
    bp.second->ws = dev_ptr;
    bp.second->ws_size = s.local_ws;
  }
  s.stage = s.stage_bytes ? static_cast<char*>(dev_ptr) + s.local_ws : nullptr;
  int* const rows_at = s.row_table.empty() ? nullptr : reinterpret_cast<int*>(static_cast<char*>(dev_ptr) + s.rows_off);
  if (rows_at && rows_at == s.rows_dev) return STENCIL_OK;  // same workspace: the lists are there
  s.rows_dev = nullptr;
  if (rows_at) {  // the needed-state lists, uploaded once per workspace (a synchronous copy)
    s.rows_dev = rows_at;
    const cudaError_t e = cudaMemcpy(s.rows_dev, s.row_table.data(), s.row_table.size() * sizeof(int),
                                     cudaMemcpyHostToDevice);
    if (e != cudaSuccess)
      return fail(STENCIL_E_CUDA, std::string("stencil_plan_set_workspace: halo row lists: ") + cudaGetErrorString(e));
  }
  return STENCIL_OK;
}

// One halo exchange of both ping-pong buffers on the communication stream: my first / last G
// owned indices go to rank -1 / rank +1, their owned indices land in my ghost indices.  A
// partition of dimension 0 sends contiguous planes; a deeper one is strided (n_outer blocks of
// G lines, local_n lines apart) and goes through the staging area: packed by 2-D copies, sent,
// received, unpacked -- all on the communication stream.
static stencil_status exchange(DistState& s, int64_t k, void* const* bufs, cudaStream_t stream) {
  NcclApi* a = s.emulate_copies ? nullptr : nccl_api();
  if (!a && !s.emulate_copies) return fail(STENCIL_E_NCCL, "NCCL unavailable");
  const DistLayout& L = s.lay;
  const int64_t G = L.ghost, local_n = L.loc_hi - L.loc_lo;
  const size_t chunk = (size_t)G * s.line_bytes;  // one outer block of a halo
  const size_t n = chunk * (size_t)s.n_outer;     // one halo (staging slot size)
  // rows of buffer b this exchange moves (all, or the needed-state list of launch k)
  const bool listed = s.rows_dev != nullptr && k >= 1 && (size_t)(2 * (k - 1) + 1) < s.row_span.size();
  auto nrows = [&](int b) { return listed ? (size_t)s.row_span[2 * (k - 1) + b].second : (size_t)s.n_outer; };
  auto rows = [&](int b) -> const int* { return listed ? s.rows_dev + s.row_span[2 * (k - 1) + b].first : nullptr; };
  auto msg = [&](int b) { return chunk * nrows(b); };
  const size_t pitch = (size_t)local_n * s.line_bytes;
  const bool strided = s.n_outer > 1;
  if (strided && !s.stage) return fail(STENCIL_E_INVALID, "stencil_run: workspace not set (halo staging)");
  ncclComm_t comm = static_cast<ncclComm_t>(s.comm);
  cudaStream_t cs = s.comm_stream;
  cudaError_t e = cudaEventRecord(s.ev_ready, stream);
  if (e == cudaSuccess) e = cudaStreamWaitEvent(cs, s.ev_ready, 0);
  if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: halo ordering: ") + cudaGetErrorString(e));
  const int64_t own0 = L.own_lo - L.loc_lo, own1 = L.own_hi - L.loc_lo;  // local indices
  const bool lo_nb = L.rank > 0, hi_nb = L.rank < L.nranks - 1;
  // staging layout per buffer b: [send lo][send hi][recv lo][recv hi]
  auto stg = [&](int b, int slot) { return s.stage + ((size_t)b * 4 + slot) * n; };
  auto at = [&](int b, int64_t idx) { return static_cast<char*>(bufs[b]) + (size_t)idx * s.line_bytes; };
  // strided halos: one gather launch for every region of this exchange (kernels/halo.cu)
  if (strided) {
    HaloCopyArgs pk{};
    for (int b = 0; b < 2; ++b) {
      if (nrows(b) == 0) continue;
      if (lo_nb) pk.reg[pk.n++] = HaloRegion{stg(b, 0), at(b, own0), chunk, pitch, chunk, nrows(b), rows(b), nullptr};
      if (hi_nb) pk.reg[pk.n++] = HaloRegion{stg(b, 1), at(b, own1 - G), chunk, pitch, chunk, nrows(b), rows(b), nullptr};
    }
    e = launch_halo_copy(pk, cs);
    if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: halo pack: ") + cudaGetErrorString(e));
  }
  if (s.emulate_copies) {  // single-GPU projection: the wire is a device-local copy
    for (int b = 0; b < 2 && e == cudaSuccess; ++b) {
      if (lo_nb && msg(b))
        e = cudaMemcpyAsync(strided ? stg(b, 2) : at(b, own0 - G), strided ? stg(b, 0) : at(b, own0), msg(b),
                            cudaMemcpyDeviceToDevice, cs);
      if (hi_nb && msg(b) && e == cudaSuccess)
        e = cudaMemcpyAsync(strided ? stg(b, 3) : at(b, own1), strided ? stg(b, 1) : at(b, own1 - G), msg(b),
                            cudaMemcpyDeviceToDevice, cs);
    }
  }
  ncclResult_t r = s.emulate_copies ? ncclSuccess : a->GroupStart();
  if (r != ncclSuccess) return nccl_fail(a, r, "ncclGroupStart");
  for (int b = 0; b < 2 && !s.emulate_copies; ++b) {
    if (msg(b) == 0) continue;
    if (lo_nb) {
      a->Send(strided ? stg(b, 0) : at(b, own0), msg(b), ncclChar, L.rank - 1, comm, cs);
      a->Recv(strided ? stg(b, 2) : at(b, own0 - G), msg(b), ncclChar, L.rank - 1, comm, cs);
    }
    if (hi_nb) {
      a->Send(strided ? stg(b, 1) : at(b, own1 - G), msg(b), ncclChar, L.rank + 1, comm, cs);
      a->Recv(strided ? stg(b, 3) : at(b, own1), msg(b), ncclChar, L.rank + 1, comm, cs);
    }
  }
  r = s.emulate_copies ? ncclSuccess : a->GroupEnd();
  if (r != ncclSuccess) return nccl_fail(a, r, "ncclGroupEnd");
  if (strided) {
    HaloCopyArgs uk{};
    for (int b = 0; b < 2; ++b) {
      if (nrows(b) == 0) continue;
      if (lo_nb) uk.reg[uk.n++] = HaloRegion{at(b, own0 - G), stg(b, 2), pitch, chunk, chunk, nrows(b), nullptr, rows(b)};
      if (hi_nb) uk.reg[uk.n++] = HaloRegion{at(b, own1), stg(b, 3), pitch, chunk, chunk, nrows(b), nullptr, rows(b)};
    }
    e = launch_halo_copy(uk, cs);
    if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: halo unpack: ") + cudaGetErrorString(e));
  }
  e = cudaEventRecord(s.ev_done, cs);
  if (e == cudaSuccess) e = cudaStreamWaitEvent(stream, s.ev_done, 0);
  if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: halo ordering: ") + cudaGetErrorString(e));
  if (a && a->CommGetAsyncError && comm) {
    ncclResult_t ae = ncclSuccess;
    if (a->CommGetAsyncError(comm, &ae) == ncclSuccess && ae != ncclSuccess && ae != ncclInProgress)
      return nccl_fail(a, ae, "NCCL async error");
  }
  return STENCIL_OK;
}

// pre_launch hook of the local plan: refresh both buffers' ghost planes
// The device-initiated exchange before launch k: my halo lines go straight into the neighbours'
// receive areas (slot k % 2) by a kernel whose last block publishes the sequence number into
// their flags; a second kernel waits for my neighbours' sequence numbers and scatters my receive
// area into my ghost lines.  Both on the compute stream (no host synchronisation, no NCCL call).
static stencil_status exchange_p2p(DistState& s, int64_t k, void* const* bufs, cudaStream_t stream) {
  const DistLayout& L = s.lay;
  if (s.loopback && (!s.peer_recv[0] && L.rank > 0 || !s.peer_recv[1] && L.rank < L.nranks - 1)) {
    std::lock_guard<std::mutex> lk(g_loop_mu);  // resolve the neighbours of this process
    auto& v = g_loop[s.group];
    if (L.rank > 0 && (int)v.size() > L.rank - 1 && v[L.rank - 1]) s.peer_recv[0] = v[L.rank - 1]->recv;
    if (L.rank < L.nranks - 1 && (int)v.size() > L.rank + 1 && v[L.rank + 1]) s.peer_recv[1] = v[L.rank + 1]->recv;
  }
  const bool lo_nb = L.rank > 0, hi_nb = L.rank < L.nranks - 1;
  if ((lo_nb && !s.peer_recv[0]) || (hi_nb && !s.peer_recv[1]))
    return fail(STENCIL_E_INVALID, "stencil_run: a neighbour's receive area is unknown (every rank's plan must exist)");
  const int64_t G = L.ghost, local_n = L.loc_hi - L.loc_lo;
  const size_t chunk = (size_t)G * s.line_bytes;
  const size_t pitch = (size_t)local_n * s.line_bytes;
  const bool listed = s.rows_dev != nullptr && k >= 1 && (size_t)(2 * (k - 1) + 1) < s.row_span.size();
  auto nrows = [&](int b) { return listed ? (size_t)s.row_span[2 * (k - 1) + b].second : (size_t)s.n_outer; };
  auto rows = [&](int b) -> const int* { return listed ? s.rows_dev + s.row_span[2 * (k - 1) + b].first : nullptr; };
  const int slot = (int)(k & 1);
  auto area = [&](char* base, int side, int b) { return base + ((size_t)(slot * 2 + side) * 2 + b) * s.recv_halo; };
  auto at = [&](int b, int64_t idx) { return static_cast<char*>(bufs[b]) + (size_t)idx * s.line_bytes; };
  const int own0 = (int)(L.own_lo - L.loc_lo), own1 = (int)(L.own_hi - L.loc_lo);
  const int seq = (int)(s.runs * (int64_t)(s.lay.n_blocks + 1) + k);
  const int blocks = halo_blocks();
  HaloCopyArgs snd{};
  HaloSignal sig{};
  for (int b = 0; b < 2; ++b) {
    if (nrows(b) == 0) continue;
    // I am my lower neighbour's upper neighbour (its side 1), and my upper neighbour's side 0
    if (lo_nb) snd.reg[snd.n++] = HaloRegion{area(s.peer_recv[0], 1, b), at(b, own0), chunk, pitch, chunk, nrows(b), rows(b), nullptr};
    if (hi_nb) snd.reg[snd.n++] = HaloRegion{area(s.peer_recv[1], 0, b), at(b, own1 - G), chunk, pitch, chunk, nrows(b), rows(b), nullptr};
  }
  if (s.emulate) {  // self-loop projection: publish exactly the flags this rank waits for
    if (lo_nb) sig.flag[sig.n++] = reinterpret_cast<int*>(s.recv + s.flag_off) + 0;
    if (hi_nb) sig.flag[sig.n++] = reinterpret_cast<int*>(s.recv + s.flag_off) + 1;
  } else {
    if (lo_nb) sig.flag[sig.n++] = reinterpret_cast<int*>(s.peer_recv[0] + s.flag_off) + 1;
    if (hi_nb) sig.flag[sig.n++] = reinterpret_cast<int*>(s.peer_recv[1] + s.flag_off) + 0;
  }
  sig.done = reinterpret_cast<unsigned int*>(s.recv + s.flag_off + 64);
  sig.done_base = s.done_count;
  sig.seq = seq;
  s.done_count += (unsigned int)blocks;
  cudaError_t e = launch_halo_send(snd, sig, blocks, stream);
  if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: halo send: ") + cudaGetErrorString(e));
  HaloCopyArgs rcv{};
  HaloWait w{};
  for (int b = 0; b < 2; ++b) {
    if (nrows(b) == 0) continue;
    if (lo_nb) rcv.reg[rcv.n++] = HaloRegion{at(b, own0 - G), area(s.recv, 0, b), pitch, chunk, chunk, nrows(b), nullptr, rows(b)};
    if (hi_nb) rcv.reg[rcv.n++] = HaloRegion{at(b, own1), area(s.recv, 1, b), pitch, chunk, chunk, nrows(b), nullptr, rows(b)};
  }
  if (lo_nb) w.flag[w.n++] = reinterpret_cast<const int*>(s.recv + s.flag_off) + 0;
  if (hi_nb) w.flag[w.n++] = reinterpret_cast<const int*>(s.recv + s.flag_off) + 1;
  w.seq = seq;
  e = launch_halo_recv(rcv, w, blocks, stream);
  if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: halo receive: ") + cudaGetErrorString(e));
  return STENCIL_OK;
}

// The fused exchange at the boundary before launch k.  Receive-area layout: mirror [side: from
// lower, from upper][buffer parity][z][G lines][x] (each side's zone of the neighbour's state),
// then the flags sent_from[lower, upper], scattered_from[lower, upper].
//   k = 0: (after the previous run's last boundary has been consumed) seed the neighbours'
//          mirrors with my send zones of both buffers;
//   k > 0: my launch k-1 has stored into their mirrors: signal "sent", wait for theirs, scatter
//          my mirror's needed rows into my ghost lines, signal "scattered", wait for theirs (they
//          no longer read the mirrors my launch k will write).
static void resolve_loop_peers(DistState& s) {
  const DistLayout& L = s.lay;
  if (!s.loopback || s.emulate) return;  // loopback: the neighbours are plans of this process
  std::lock_guard<std::mutex> lk(g_loop_mu);
  auto& v = g_loop[s.group];
  if (L.rank > 0 && !s.peer_recv[0] && (int)v.size() > L.rank - 1 && v[L.rank - 1]) s.peer_recv[0] = v[L.rank - 1]->recv;
  if (L.rank < L.nranks - 1 && !s.peer_recv[1] && (int)v.size() > L.rank + 1 && v[L.rank + 1])
    s.peer_recv[1] = v[L.rank + 1]->recv;
}

static stencil_status exchange_fused(DistState& s, int64_t k, void* const* bufs, cudaStream_t stream) {
  const DistLayout& L = s.lay;
  resolve_loop_peers(s);
  const bool lo_nb = L.rank > 0, hi_nb = L.rank < L.nranks - 1;
  if ((lo_nb && !s.peer_recv[0]) || (hi_nb && !s.peer_recv[1]))
    return fail(STENCIL_E_INVALID, "stencil_run: a neighbour's receive area is unknown (every rank's plan must exist)");
  const int64_t G = L.ghost, local_n = L.loc_hi - L.loc_lo;
  const size_t chunk = (size_t)G * s.line_bytes, pitch = (size_t)local_n * s.line_bytes;
  const size_t M = chunk * (size_t)s.n_outer;  // one parity of one side's mirror
  auto mirror = [&](char* base, int side, int b) { return base + ((size_t)side * 2 + b) * M; };
  auto flags = [&](char* base) { return reinterpret_cast<int*>(base + s.flag_off); };
  auto at = [&](int b, int64_t idx) { return static_cast<char*>(bufs[b]) + (size_t)idx * s.line_bytes; };
  const int own0 = (int)(L.own_lo - L.loc_lo), own1 = (int)(L.own_hi - L.loc_lo);
  const int seq = (int)(s.runs * (int64_t)(s.lay.n_blocks + 1) + k);
  const int blocks = halo_blocks();
  // flag word `idx` of my neighbour on side `nb_side` that refers to me (self-loop projection:
  // the word of mine I will wait on)
  auto remote = [&](int nb_side, int idx_base) -> int* {
    if (s.emulate) return flags(s.recv) + idx_base + nb_side;
    return flags(s.peer_recv[nb_side]) + idx_base + (1 - nb_side);
  };
  auto wait = [&](int idx_base, int sq) -> cudaError_t {
    HaloCopyArgs none{};
    HaloWait w{};
    if (lo_nb) w.flag[w.n++] = flags(s.recv) + idx_base + 0;
    if (hi_nb) w.flag[w.n++] = flags(s.recv) + idx_base + 1;
    w.seq = sq;
    return launch_halo_recv(none, w, blocks, stream);
  };
  auto signal = [&](int idx_base) -> cudaError_t {
    int* f[2];
    int n = 0;
    if (lo_nb) f[n++] = remote(0, idx_base);
    if (hi_nb) f[n++] = remote(1, idx_base);
    return launch_halo_signal(n, f, seq, stream);
  };
  cudaError_t e = cudaSuccess;
  if (k == 0) {
    if (s.runs > 0) e = wait(2, seq - 2);  // the neighbours scattered the previous run's last data
    HaloCopyArgs cp{};
    for (int b = 0; b < 2 && e == cudaSuccess; ++b) {
      char* lo_dst = s.emulate ? mirror(s.recv, 0, b) : (lo_nb ? mirror(s.peer_recv[0], 1, b) : nullptr);
      char* hi_dst = s.emulate ? mirror(s.recv, 1, b) : (hi_nb ? mirror(s.peer_recv[1], 0, b) : nullptr);
      if (lo_nb) cp.reg[cp.n++] = HaloRegion{lo_dst, at(b, own0), chunk, pitch, chunk, (size_t)s.n_outer, nullptr, nullptr};
      if (hi_nb) cp.reg[cp.n++] = HaloRegion{hi_dst, at(b, own1 - G), chunk, pitch, chunk, (size_t)s.n_outer, nullptr, nullptr};
    }
    if (e == cudaSuccess) e = launch_halo_copy(cp, stream);
  } else {
    const bool listed = s.rows_dev != nullptr && (size_t)(2 * (k - 1) + 1) < s.row_span.size();
    auto nrows = [&](int b) { return listed ? (size_t)s.row_span[2 * (k - 1) + b].second : (size_t)s.n_outer; };
    auto rows = [&](int b) -> const int* { return listed ? s.rows_dev + s.row_span[2 * (k - 1) + b].first : nullptr; };
    e = signal(0);
    if (e == cudaSuccess) e = wait(0, seq);
    HaloCopyArgs sc{};
    for (int b = 0; b < 2; ++b) {
      if (nrows(b) == 0) continue;
      if (lo_nb) sc.reg[sc.n++] = HaloRegion{at(b, own0 - G), mirror(s.recv, 0, b), pitch, chunk, chunk, nrows(b), rows(b), rows(b)};
      if (hi_nb) sc.reg[sc.n++] = HaloRegion{at(b, own1), mirror(s.recv, 1, b), pitch, chunk, chunk, nrows(b), rows(b), rows(b)};
    }
    if (e == cudaSuccess) e = launch_halo_copy(sc, stream);
    if (e == cudaSuccess) e = signal(2);
    if (e == cudaSuccess) e = wait(2, seq);
  }
  if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("stencil_run: fused halo exchange: ") + cudaGetErrorString(e));
  return STENCIL_OK;
}

static stencil_status ghost_hook(void* ctx, int64_t k, void* const* bufs, void* stream) {
  DistState& s = *static_cast<DistState*>(ctx);
  if (s.lay.nranks <= 1 || (s.emulate && !s.emulate_copies)) return STENCIL_OK;
  if (s.fused) return exchange_fused(s, k, bufs, static_cast<cudaStream_t>(stream));
  if (k == 0) return STENCIL_OK;  // (the other paths exchange before launches k >= 1 only)
  if (s.p2p) return exchange_p2p(s, k, bufs, static_cast<cudaStream_t>(stream));
  return exchange(s, k, bufs, static_cast<cudaStream_t>(stream));
}

stencil_status run_dist(Plan& p, const void* const* in, void* const* out, void* stream_) {
  DistState& s = *p.dist;
  cudaStream_t stream = static_cast<cudaStream_t>(stream_);
  if (!in || !out || !in[0] || !out[0]) return fail(STENCIL_E_INVALID, "stencil_run: NULL field pointer");
  if ((reinterpret_cast<uintptr_t>(in[0]) | reinterpret_cast<uintptr_t>(out[0])) % 16)
    return fail(STENCIL_E_INVALID, "stencil_run: field pointers must be 16-B aligned");
  int dev = -1;
  if (cudaGetDevice(&dev) != cudaSuccess || dev != s.comm_dev)
    return fail(STENCIL_E_CUDA, "stencil_run: a distributed plan runs on the device it was created on");
  Plan* lp = s.bplans.empty() ? nullptr : s.bplans[0].second;
  if (!lp) return STENCIL_OK;
  lp->pre_launch = ghost_hook;
  lp->pre_launch_ctx = &s;
  lp->mir[0] = lp->mir[1] = nullptr;
  lp->mir_G = 0;
  resolve_loop_peers(s);
  static const bool no_store = std::getenv("HEXS_DIST_FUSED_NOSTORE") && std::atoi(std::getenv("HEXS_DIST_FUSED_NOSTORE"));
  if (s.fused && s.lay.nranks > 1 && !no_store) {  // the phase kernel mirrors its send zones (local lines)
    const size_t M = (size_t)s.lay.ghost * s.line_bytes * (size_t)s.n_outer;
    const bool lo_nb = s.lay.rank > 0, hi_nb = s.lay.rank < s.lay.nranks - 1;
    char* lo_base = s.emulate ? s.recv : s.peer_recv[0];
    char* hi_base = s.emulate ? s.recv : s.peer_recv[1];
    if (lo_nb && lo_base) lp->mir[0] = lo_base + (s.emulate ? 0 : 2 * M);   // the lower neighbour's side 1
    if (hi_nb && hi_base) lp->mir[1] = hi_base + (s.emulate ? 2 * M : 0);   // the upper neighbour's side 0
    lp->mir_y0[0] = (int)(s.lay.own_lo - s.lay.loc_lo);
    lp->mir_y0[1] = (int)(s.lay.own_hi - s.lay.loc_lo - s.lay.ghost);
    lp->mir_G = (int)s.lay.ghost;
    // (HEXS_DIST_MIRFENCE=0: no system-scope fence -- measurement aid only)
    static const char* mf = std::getenv("HEXS_DIST_MIRFENCE");
    lp->mir_fence = mf ? std::atoi(mf) : 1;
  }
  // the local plan copies in -> out and runs the global launch table over the slab, exchanging
  // the ghost planes before every launch but the first
  const stencil_status st = run_plan(*lp, in, out, stream);
  if (st == STENCIL_OK) ++s.runs;
  return st;
}

}  // namespace hexs

using namespace hexs;

extern "C" {

stencil_status stencil_dist_unique_id(void* id_out) {
  clear_error();
  if (!id_out) return fail(STENCIL_E_INVALID, "stencil_dist_unique_id: NULL output");
  NcclApi* a = nccl_api();
  if (!a) return fail(STENCIL_E_NCCL, "stencil_dist_unique_id: NCCL unavailable");
  ncclUniqueId id;
  ncclResult_t r = a->GetUniqueId(&id);
  if (r != ncclSuccess) return nccl_fail(a, r, "ncclGetUniqueId");
  std::memcpy(id_out, &id, sizeof(id));
  return STENCIL_OK;
}

stencil_status stencil_dist_layout(stencil_desc_t global_desc, int64_t T_steps, const stencil_tile_t* tile,
                                   int rank, int nranks, int part_dim, stencil_dist_info_t* info) {
  clear_error();
  Desc* d = reinterpret_cast<Desc*>(global_desc);
  if (!d || d->magic != kDescMagic || !info) return fail(STENCIL_E_INVALID, "stencil_dist_layout: bad arguments");
  DistLayout L{};
  stencil_status st = dist_layout(*d, T_steps, tile, rank, nranks, part_dim, &L);
  if (st != STENCIL_OK) return st;
  stencil_dist_info_t o{};
  o.rank = L.rank;
  o.nranks = L.nranks;
  o.part_dim = L.part_dim;
  for (int q = 0; q < 3; ++q) {
    o.global_ext[q] = q < d->dims ? d->ext[q] : 1;
    o.local_ext[q] = o.global_ext[q];
  }
  o.local_ext[L.part_dim] = L.loc_hi - L.loc_lo;
  o.own_lo = L.own_lo;
  o.own_hi = L.own_hi;
  o.loc_lo = L.loc_lo;
  o.loc_hi = L.loc_hi;
  o.ghost = L.ghost;
  o.time_block = L.time_block;
  o.n_blocks = L.n_blocks;
  o.h = L.h;
  o.ghost_fraction = L.ghost_fraction;
  *info = o;
  return STENCIL_OK;
}

stencil_status stencil_plan_dist(stencil_plan_t* out, stencil_desc_t global_desc, int64_t T_steps,
                                 const stencil_tile_t* tile, const void* nccl_unique_id, int rank, int nranks,
                                 int part_dim) {
  clear_error();
  if (!out) return fail(STENCIL_E_INVALID, "stencil_plan_dist: out is NULL");
  *out = nullptr;
  Desc* d = reinterpret_cast<Desc*>(global_desc);
  if (!d || d->magic != kDescMagic) return fail(STENCIL_E_INVALID, "stencil_plan_dist: bad descriptor");
  if (!nccl_unique_id) return fail(STENCIL_E_INVALID, "stencil_plan_dist: NULL NCCL unique id");
  std::unique_ptr<DistState> s(new (std::nothrow) DistState());
  if (!s) return fail(STENCIL_E_OOM, "stencil_plan_dist: out of host memory");
  stencil_status st = dist_layout(*d, T_steps, tile, rank, nranks, part_dim, &s->lay);
  if (st != STENCIL_OK) return st;
  const DistLayout& L = s->lay;
  const int pd = L.part_dim;
  // the local slab's descriptor: same class / coefficients / dtype, extent loc_hi - loc_lo
  s->local = *d;
  s->local.ext[pd] = L.loc_hi - L.loc_lo;
  if (s->local.ext[pd] < 3) return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan_dist: local slab thinner than 3 indices");
  s->global_n = d->ext[pd];
  s->line_bytes = d->elem();
  for (int q = pd + 1; q < d->dims; ++q) s->line_bytes *= (size_t)d->ext[q];
  s->n_outer = 1;
  for (int q = 0; q < pd; ++q) s->n_outer *= d->ext[q];
  s->blocks.push_back(T_steps);
  const stencil_tile_t lt = dist_local_tile(*d, tile, nranks);
  {
    // the local plan: the global schedule restricted to the slab (hexagon rows translated by
    // loc_lo when the partitioned dimension is the hexagonal one, so the tiling matches the
    // global one)
    Plan* probe = nullptr;
    st = build_plan(s->local, T_steps, &lt, &probe);
    if (st != STENCIL_OK) return st;
    const int64_t origin = probe->hd == pd ? L.loc_lo : 0;
    delete probe;
    Plan* bp = nullptr;
    st = build_plan(s->local, T_steps, &lt, &bp, origin);
    if (st != STENCIL_OK) return st;
    if (bp->h != L.h) {
      delete bp;
      return fail(STENCIL_E_INVALID, "stencil_plan_dist: local tile differs from the layout's");
    }
    s->lay.n_blocks = (int64_t)bp->launches.size();
    s->bplans.push_back({T_steps, bp});
  }
  // NCCL communicator and the communication stream on the current device
  if (cudaGetDevice(&s->comm_dev) != cudaSuccess) return fail(STENCIL_E_CUDA, "stencil_plan_dist: no CUDA device");
  if (cudaStreamCreateWithFlags(&s->comm_stream, cudaStreamNonBlocking) != cudaSuccess ||
      cudaEventCreateWithFlags(&s->ev_ready, cudaEventDisableTiming) != cudaSuccess ||
      cudaEventCreateWithFlags(&s->ev_done, cudaEventDisableTiming) != cudaSuccess)
    return fail(STENCIL_E_CUDA, "stencil_plan_dist: stream / event creation failed");
  // HEXS_DIST_EMULATE=1: one process plays one rank of nranks on its own GPU -- no
  // communicator, no exchanges (the ghost planes keep their initial values, so results are not
  // the global ones); it measures a rank's compute for scaling projections on a single GPU
  s->emulate = std::getenv("HEXS_DIST_EMULATE") && std::atoi(std::getenv("HEXS_DIST_EMULATE")) != 0;
  // =2: plus the NCCL path's halo copies (a device-local copy as the wire); =3: plus the
  // device-initiated path's kernels, the rank's own receive area standing in for its neighbours'
  const int emu_mode = s->emulate ? std::atoi(std::getenv("HEXS_DIST_EMULATE")) : 0;
  s->emulate_copies = emu_mode >= 2;
  // HEXS_DIST_LOOPBACK=1: the ranks are plans of ONE process on one device (no communicator; the
  // device-initiated exchange between them) -- the single-GPU test of the multi-rank protocol
  s->loopback = !s->emulate && std::getenv("HEXS_DIST_LOOPBACK") && std::atoi(std::getenv("HEXS_DIST_LOOPBACK")) != 0;
  if (!s->emulate && !s->loopback) {  // (also for one rank: the same NCCL bootstrap path, no exchange ever runs)
    NcclApi* a = nccl_api();
    if (!a) return fail(STENCIL_E_NCCL, "stencil_plan_dist: NCCL unavailable");
    ncclUniqueId id;
    std::memcpy(&id, nccl_unique_id, sizeof(id));
    ncclComm_t comm = nullptr;
    ncclResult_t r = a->CommInitRank(&comm, nranks, id, rank);
    if (r != ncclSuccess) return nccl_fail(a, r, "ncclCommInitRank");
    s->comm = comm;
  }
  // the dist plan itself: the primary block plan's schedule, the whole run's step count
  Plan* p = new (std::nothrow) Plan();
  if (!p) return fail(STENCIL_E_OOM, "stencil_plan_dist: out of host memory");
  Plan* primary = s->plan_for(s->blocks.empty() ? 0 : s->blocks[0]);
  if (primary) {
    p->desc = primary->desc;
    p->hd = primary->hd;
    p->h = primary->h;
    p->w0 = primary->w0;
  } else {
    p->desc = s->local;
  }
  p->T_steps = T_steps;
  p->tau_levels = T_steps * (int64_t)d->stmts.size();
  p->executor = primary ? primary->executor : EXEC_GENERIC;
  size_t ws = 0;
  for (auto& bp : s->bplans) ws = std::max(ws, bp.second->ws_bytes);
  s->local_ws = (ws + 255) / 256 * 256;
  // Device-initiated exchange (default for nranks > 1; HEXS_DIST_P2P=0 keeps NCCL send/recv):
  // a receive area in NCCL symmetric memory (ncclMemAlloc + ncclCommWindowRegister, collective),
  // whose neighbours' views are the window's LSA pointers; loopback mode: cudaMalloc and the
  // process-local registry.  Halo copies move 16-B units: chunk and pitch must be 16-B multiples.
  {
    const char* pe = std::getenv("HEXS_DIST_P2P");
    const bool want = nranks > 1 && !(pe && std::atoi(pe) == 0) && (!s->emulate || emu_mode == 3);
    const size_t chunk = (size_t)L.ghost * s->line_bytes;
    if (want && s->line_bytes % 16 == 0) {  // (rank-independent: every chunk and pitch 16-B granular)
      s->recv_halo = (chunk * (size_t)s->n_outer + 255) / 256 * 256;
      s->flag_off = 8 * s->recv_halo;
      s->recv_bytes = s->flag_off + 256;
      if (emu_mode == 3) {  // self-loop: measures the send / wait / scatter kernels of one rank
        void* r = nullptr;
        if (cudaMalloc(&r, s->recv_bytes) != cudaSuccess || cudaMemset(r, 0, s->recv_bytes) != cudaSuccess)
          return fail(STENCIL_E_OOM, "stencil_plan_dist: emulated receive area");
        s->recv = static_cast<char*>(r);
        s->loopback = true;  // (freed with cudaFree; no registry entry: group stays empty)
        s->peer_recv[0] = s->peer_recv[1] = s->recv;
        s->p2p = true;
      } else if (s->loopback) {
        void* r = nullptr;
        if (cudaMalloc(&r, s->recv_bytes) != cudaSuccess || cudaMemset(r, 0, s->recv_bytes) != cudaSuccess)
          return fail(STENCIL_E_OOM, "stencil_plan_dist: loopback receive area");
        s->recv = static_cast<char*>(r);
        s->group.assign(static_cast<const char*>(nccl_unique_id), 128);
        std::lock_guard<std::mutex> lk(g_loop_mu);
        auto& v = g_loop[s->group];
        if ((int)v.size() < nranks) v.resize(nranks, nullptr);
        v[rank] = s.get();
        s->p2p = true;
      } else if (NcclApi* a = nccl_api()) {
        // every rank must take the same path (the window registration is collective): each step's
        // local outcome is min-reduced over the communicator before the next
        auto all_ok = [&](int ok) {
          if (!s->comm || !a->AllReduce) return false;
          int* dv = nullptr;
          if (cudaMalloc(reinterpret_cast<void**>(&dv), sizeof(int)) != cudaSuccess) return false;
          bool good = cudaMemcpy(dv, &ok, sizeof(int), cudaMemcpyHostToDevice) == cudaSuccess &&
                      a->AllReduce(dv, dv, 1, ncclInt32, ncclMin, static_cast<ncclComm_t>(s->comm), s->comm_stream) ==
                          ncclSuccess &&
                      cudaStreamSynchronize(s->comm_stream) == cudaSuccess &&
                      cudaMemcpy(&ok, dv, sizeof(int), cudaMemcpyDeviceToHost) == cudaSuccess;
          cudaFree(dv);
          return good && ok == 1;
        };
        void* r = nullptr;
        const bool have = a->MemAlloc && a->WindowRegister && a->WindowDeregister && a->MemFree;
        bool ok = have && a->MemAlloc(&r, s->recv_bytes) == ncclSuccess && r &&
                  cudaMemset(r, 0, s->recv_bytes) == cudaSuccess;
        if (r) s->recv = static_cast<char*>(r);
        if (all_ok(ok ? 1 : 0)) {
          ncclWindow_t w = nullptr;
          ok = a->WindowRegister(static_cast<ncclComm_t>(s->comm), r, s->recv_bytes, &w, NCCL_WIN_COLL_SYMMETRIC) ==
                   ncclSuccess &&
               w;
          if (w) s->win = w;
          void* pp = nullptr;
          if (ok && rank > 0) {
            ok = halo_peer_pointer(w, rank - 1, &pp, s->comm_stream) == cudaSuccess && pp;
            s->peer_recv[0] = static_cast<char*>(pp);
          }
          if (ok && rank < nranks - 1) {
            ok = halo_peer_pointer(w, rank + 1, &pp, s->comm_stream) == cudaSuccess && pp;
            s->peer_recv[1] = static_cast<char*>(pp);
          }
          s->p2p = all_ok(ok ? 1 : 0);
        }
        if (!s->p2p) s->release_p2p();  // fall back to ncclSend / ncclRecv
      }
    }
    if (s->loopback && !s->p2p && nranks > 1)
      return fail(STENCIL_E_UNSUPPORTED, "stencil_plan_dist: loopback mode needs 16-B aligned halos");
  }
  // strided partitions exchanged by NCCL send/recv: staging for both buffers' 2 send + 2 receive halos
  s->stage_bytes = !s->p2p && s->n_outer > 1 && nranks > 1 ? 8 * (size_t)L.ghost * s->line_bytes * (size_t)s->n_outer : 0;
  // needed-state row lists: the hexagonal dimension 0 whole (its coordinate is the outer index
  // of the halo blocks), a classical dimension partitioned
  Plan* lp0 = s->bplans.empty() ? nullptr : s->bplans[0].second;
  if ((s->stage_bytes || (s->p2p && s->n_outer > 1)) && lp0 && halo_rows_table(*lp0, pd, s->row_table, s->row_span)) {
    s->rows_off = s->local_ws + s->stage_bytes;
    s->rows_bytes = (s->row_table.size() * sizeof(int) + 255) / 256 * 256;
  }
  p->ws_bytes = s->local_ws + s->stage_bytes + s->rows_bytes;
  // fused halo stores (HEXS_DIST_FUSED=1, opt-in): the 3D tile-wavefront kernel on y slabs of at
  // least 2G lines (rank-independent test: the smallest slab).  Measured: its
  // mirror-storing instantiation runs ~15 % slower than the plain kernel, which eats the overlap
  // it buys, so the separate device-initiated exchange stays the default
  {
    const char* fe = std::getenv("HEXS_DIST_FUSED");
    s->fused = s->p2p && lp0 && lp0->executor == EXEC_FAST3D && pd == 1 && lp0->hd == 0 &&
               d->ext[pd] / nranks >= 2 * L.ghost && fe && std::atoi(fe) != 0;
  }
  p->dist = s.release();
  *out = reinterpret_cast<stencil_plan_t>(p);
  return STENCIL_OK;
}

stencil_status stencil_dist_local_plan(stencil_plan_t* out, stencil_desc_t global_desc, int64_t T_steps,
                                       const stencil_tile_t* tile, int rank, int nranks, int part_dim) {
  clear_error();
  if (!out) return fail(STENCIL_E_INVALID, "stencil_dist_local_plan: out is NULL");
  *out = nullptr;
  Desc* d = reinterpret_cast<Desc*>(global_desc);
  if (!d || d->magic != kDescMagic) return fail(STENCIL_E_INVALID, "stencil_dist_local_plan: bad descriptor");
  DistLayout L{};
  stencil_status st = dist_layout(*d, T_steps, tile, rank, nranks, part_dim, &L);
  if (st != STENCIL_OK) return st;
  Desc local = *d;
  local.ext[L.part_dim] = L.loc_hi - L.loc_lo;
  if (local.ext[L.part_dim] < 3) return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_dist_local_plan: slab thinner than 3 indices");
  const stencil_tile_t lt = dist_local_tile(*d, tile, nranks);
  Plan* probe = nullptr;
  st = build_plan(local, T_steps, &lt, &probe);
  if (st != STENCIL_OK) return st;
  const int64_t origin = probe->hd == L.part_dim ? L.loc_lo : 0;
  delete probe;
  Plan* p = nullptr;
  st = build_plan(local, T_steps, &lt, &p, origin);
  if (st != STENCIL_OK) return st;
  *out = reinterpret_cast<stencil_plan_t>(p);
  return STENCIL_OK;
}

stencil_status stencil_dist_halo_rows(stencil_plan_t local_plan, int part_dim, int64_t k, int buffer, int32_t* rows,
                                     int64_t cap, int64_t* n) {
  clear_error();
  Plan* p = as_plan(local_plan);
  if (!p || p->dist || !n || buffer < 0 || buffer > 1 || k < 1)
    return fail(STENCIL_E_INVALID, "stencil_dist_halo_rows: bad arguments");
  std::vector<int> table;
  std::vector<std::pair<int64_t, int64_t>> span;
  if (!halo_rows_table(*p, part_dim, table, span)) {
    *n = -1;  // the rule does not apply: every outer row travels
    return STENCIL_OK;
  }
  if ((size_t)(2 * (k - 1) + buffer) >= span.size()) return fail(STENCIL_E_INVALID, "stencil_dist_halo_rows: k out of range");
  const auto sp = span[2 * (k - 1) + buffer];
  *n = sp.second;
  if (rows)
    for (int64_t i = 0; i < sp.second && i < cap; ++i) rows[i] = table[sp.first + i];
  return STENCIL_OK;
}

stencil_status stencil_dist_info(stencil_plan_t plan, stencil_dist_info_t* info) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !p->dist || !info) return fail(STENCIL_E_INVALID, "stencil_dist_info: not a distributed plan");
  const DistState& s = *p->dist;
  const DistLayout& L = s.lay;
  stencil_dist_info_t o{};
  o.rank = L.rank;
  o.nranks = L.nranks;
  o.part_dim = L.part_dim;
  for (int q = 0; q < 3; ++q) o.local_ext[q] = o.global_ext[q] = q < s.local.dims ? s.local.ext[q] : 1;
  o.global_ext[L.part_dim] = s.global_n;
  o.local_ext[L.part_dim] = L.loc_hi - L.loc_lo;
  o.own_lo = L.own_lo;
  o.own_hi = L.own_hi;
  o.loc_lo = L.loc_lo;
  o.loc_hi = L.loc_hi;
  o.ghost = L.ghost;
  o.time_block = L.time_block;
  o.n_blocks = L.n_blocks;
  o.h = L.h;
  o.ghost_fraction = L.ghost_fraction;
  int64_t launches = 0;
  for (int64_t len : s.blocks) {
    const Plan* bp = s.plan_for(len);
    launches += bp->executor == EXEC_NAIVE ? bp->tau_levels : (int64_t)bp->launches.size();
  }
  o.launches_per_run = launches;
  o.exchange = L.nranks <= 1 || (s.emulate && !s.emulate_copies) ? STENCIL_EXCHANGE_NONE
               : s.fused                                        ? STENCIL_EXCHANGE_FUSED
               : s.p2p                                          ? STENCIL_EXCHANGE_P2P
                                                                : STENCIL_EXCHANGE_NCCL;
  *info = o;
  return STENCIL_OK;
}

stencil_status stencil_dist_block_plan(stencil_plan_t plan, int index, stencil_plan_t* block) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !p->dist || !block) return fail(STENCIL_E_INVALID, "stencil_dist_block_plan: not a distributed plan");
  if (index < 0 || index >= (int)p->dist->bplans.size())
    return fail(STENCIL_E_INVALID, "stencil_dist_block_plan: index out of range");
  *block = reinterpret_cast<stencil_plan_t>(p->dist->bplans[index].second);
  return STENCIL_OK;
}

}  // extern "C"

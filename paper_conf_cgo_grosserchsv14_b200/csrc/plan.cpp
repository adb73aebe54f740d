// plan.cpp -- tile-parameter validation (a2) and the hybrid schedule -> launch table (a3).
//
// Implements Sec. 3.3-3.6 of the paper for the planner:
//   cone slopes delta0/delta1 along the hexagonal dimension  (Sec. 3.3.2, Fig. 3)
//   width bound, eq. (1)
//   two-phase tile schedule, eqs. (2)-(5); the phase-0 numerator uses floor(delta0 h)
//   (reading R1 -- the extracted eq. (3) shows floor(delta1 h), which does not
//   tile the plane when delta0 != delta1)
//   hexagon constraints (6),(7),(8),(10),(12),(13) in local box coordinates
//
//   classical tiling eqs. (14)-(17) with u = the local box row
//   host loop "repeatedly iterating over two CUDA kernels"
#include <algorithm>
#include <cstdlib>
#include <climits>
#include <cmath>
#include <memory>
#include <new>
#include <set>
#include <string>

#include <cuda_runtime.h>

#include "internal.h"

namespace hexs {

// SMs of the current device (148 on B200 when no device is visible, e.g. planning on a host)
static int device_sm_count() {
  int dev = 0, sms = 0;
  if (cudaGetDevice(&dev) == cudaSuccess && cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) == cudaSuccess &&
      sms > 0)
    return sms;
  cudaGetLastError();
  return 148;
}

namespace {

struct Slopes {
  Rat d0, d1;
};

// delta0 = max(0, max ds/dt), delta1 = max(0, max -ds/dt) over the distance vectors
// (Delta s0 <= delta0 Delta t, Delta s0 >= -delta1 Delta t).
Slopes cone_slopes(const std::vector<std::vector<int64_t>>& dist, int dim) {
  Slopes s{make_rat(0, 1), make_rat(0, 1)};
  for (auto& v : dist) {
    Rat fwd = make_rat(v[1 + dim], v[0]);
    Rat bwd = make_rat(-v[1 + dim], v[0]);
    if (rat_less(s.d0, fwd)) s.d0 = fwd;
    if (rat_less(s.d1, bwd)) s.d1 = bwd;
  }
  return s;
}

int64_t floor_rat_mul(const Rat& r, int64_t h) { return floor_div(r.n * h, r.d); }

// eq. (1): w0 >= max(delta0 + {delta0 h}, delta1 + {delta1 h}) - 1.  Returns the smallest
// admissible integer w0.
int64_t w0_bound(const Rat& d0, const Rat& d1, int64_t h) {
  auto term = [&](const Rat& d) {
    // d + {d h} - 1 = d + (d h - floor(d h)) - 1, as a rational with denominator d.d
    int64_t num = d.n + (d.n * h - floor_rat_mul(d, h) * d.d) - d.d;
    return ceil_div(num, d.d);
  };
  return std::max<int64_t>(0, std::max(term(d0), term(d1)));
}

bool in_hexagon(const Plan& p, int64_t a, int64_t b) {
  const int64_t n0 = p.d0.n, q0 = p.d0.d, n1 = p.d1.n, q1 = p.d1.d, h = p.h, w0 = p.w0;
  // (6)  d0 a - b <= (2h+1) d0 - F0
  if (n0 * a - b * q0 > (2 * h + 1) * n0 - p.F0 * q0) return false;
  // (7)  a <= 2h+1 ; (13) a >= 0
  if (a > 2 * h + 1 || a < 0) return false;
  // (8)  d1 a + b <= (2h+1) d1 + F0 + w0
  if (n1 * a + b * q1 > (2 * h + 1) * n1 + (p.F0 + w0) * q1) return false;
  // (10) d1 a + b >= h d1 - (q1-1)/q1
  if (n1 * a + b * q1 < h * n1 - (q1 - 1)) return false;
  // (12) d0 a - b >= d0 h - F0 - w0 - F1 - (q0-1)/q0
  if (n0 * a - b * q0 < h * n0 - (p.F0 + w0 + p.F1) * q0 - (q0 - 1)) return false;
  return true;
}

void hexagon_traffic(Plan& p) {
  std::set<std::pair<int64_t, int64_t>> pts, ins;
  for (int a = 0; a < p.H; ++a)
    for (int b = p.lo[a]; b <= p.hi[a]; ++b) pts.insert({a, b});
  // offsets along the hexagonal dimension read by any statement
  std::set<int> offs;
  for (auto& st : p.desc.stmts)
    for (auto& ac : st.reads) offs.insert(ac.off[p.hd]);
  int64_t out = 0;
  for (auto& q : pts) {
    bool is_out = false;
    for (int o : offs) {
      if (!pts.count({q.first - 1, q.second + o})) ins.insert({q.first - 1, q.second + o});
      if (!pts.count({q.first + 1, q.second - o})) is_out = true;
    }
    out += is_out;
  }
  p.tile_points = (int64_t)pts.size();
  p.tile_in = (int64_t)ins.size();
  p.tile_out = out;
}

}  // namespace

bool schedule_of(const Plan& p, int64_t tau, const int64_t* s, int64_t* sched) {
  const int64_t s0 = s[p.hd];
  for (int ph = 0; ph < 2; ++ph) {
    int64_t T, n, a;
    if (ph == 0) {
      T = floor_div(tau + p.h + 1, p.H);                    // eq. (2)
      n = s0 + p.hex_origin + p.F0 + p.w0 + 1 + T * p.c;     // eq. (3), floor(d0 h)
      a = tau + p.h + 1 - T * p.H;
    } else {
      T = floor_div(tau, p.H);                               // eq. (4)
      n = s0 + p.hex_origin + T * p.c;                       // eq. (5)
      a = tau - T * p.H;
    }
    const int64_t S0 = floor_div(n, p.W), b = n - S0 * p.W;
    if (b < p.lo[a] || b > p.hi[a]) continue;
    int k = 0;
    sched[k++] = T;
    sched[k++] = ph;
    sched[k++] = S0;
    int64_t sp[2] = {0, 0};
    for (int q = 0; q < p.ncls; ++q) {
      // eqs. (14), (17) with the tile translation offset of Sec. 4.2.3
      const int64_t x = s[p.cls[q]] - p.ctrans[q] + (int64_t)p.dcls[q] * a;
      const int64_t Si = floor_div(x, p.w[q]);
      sched[k++] = Si;
      sp[q] = x - Si * p.w[q];
    }
    sched[k++] = a;
    sched[k++] = b;
    for (int q = 0; q < p.ncls; ++q) sched[k++] = sp[q];
    return true;
  }
  return false;
}

stencil_status build_plan(const Desc& d, int64_t T_steps, const stencil_tile_t* tile, Plan** out,
                          int64_t hex_origin) {
  if (T_steps < 0) return fail(STENCIL_E_INVALID, "stencil_plan: T_steps < 0");
  Plan* p = new (std::nothrow) Plan();
  if (!p) return fail(STENCIL_E_OOM, "stencil_plan: out of host memory");
  std::unique_ptr<Plan> guard(p);
  p->desc = d;
  p->T_steps = T_steps;
  p->hex_origin = hex_origin;
  p->tau_levels = T_steps * (int64_t)d.stmts.size();
  stencil_tile_t t{};
  t.hex_dim = -1;  // NULL tile: everything automatic
  if (tile) t = *tile;
  // hex_dim < 0: automatic -- the streaming 3D kernel tiles y hexagonally (its stream runs along
  // z, the outermost dimension, PAPER.md:633-641 allows any non-innermost dimension); everything
  // else tiles the outermost dimension
  const bool s3_class = d.dims == 3 && (d.kind == STENCIL_STAR3D7 || d.kind == STENCIL_GRADIENT3D) &&
                        d.dtype == STENCIL_F32 && t.flags == STENCIL_EXEC_AUTO && d.ext[2] % 4 == 0 &&
                        d.ext[2] < (int64_t(1) << 30) && d.ext[1] < (int64_t(1) << 30) &&
                        d.ext[0] < (int64_t(1) << 30);
  // (measured on B200: the tile-wavefront kernel over (t, z) is still the faster default for the
  // star classes; HEXS_STREAM3D=1 makes the streaming kernel the automatic choice)
  static const bool s3_auto = std::getenv("HEXS_STREAM3D") && std::atoi(std::getenv("HEXS_STREAM3D")) != 0;
  p->hd = t.hex_dim >= 0 ? t.hex_dim : (s3_class && s3_auto ? 1 : 0);
  if (p->hd < 0 || p->hd >= d.dims - 1)
    return fail(STENCIL_E_INVALID, "stencil_plan: hex_dim must be a non-innermost dimension (PAPER.md:636-641)");
  p->ncls = 0;
  for (int q = 0; q < d.dims; ++q)
    if (q != p->hd) p->cls[p->ncls++] = q;

  // a1: dependence analysis -> slopes
  auto dist = dependence_distances(d);
  Slopes sl = cone_slopes(dist, p->hd);
  p->d0 = sl.d0;
  p->d1 = sl.d1;
  for (int q = 0; q < p->ncls; ++q) {
    Slopes c = cone_slopes(dist, p->cls[q]);
    p->dcls[q] = (int)ceil_div(c.d1.n, c.d1.d);  // integer skew >= delta1_i (Sec. 3.4)
  }

  // a2: tile parameters
  const int flags = t.flags;
  const bool ablation = flags >= STENCIL_EXEC_T4A && flags <= STENCIL_EXEC_T4F;
  bool auto_tile = (t.h == 0 && t.w0 == 0);
  int h = t.h, w0 = t.w0;
  const int dtype = d.dtype;
  if (auto_tile) {
    if (ablation) {
      h = 2;
      w0 = 7;  // Table 4's tile
    } else if (d.kind == STENCIL_FDTD2D) {
      // 24 tau-levels = 8 full steps per tile (h+1 a multiple of 3, reading R14); w0 as
      // small as possible while every launch's hexagons (W = 2 w0 + 2 + h + h/2 rows) fit one
      // wave of the FDTD kernel (fdtd_ctas_per_sm() CTAs per SM): a second, partial wave would double the
      // launch time (grid quantisation).  Best measured on B200: profiles/round1/.
      h = 11;
      w0 = 5;
      const int64_t slots = (int64_t)fdtd_ctas_per_sm() * device_sm_count();
      auto Wof = [&](int w) { return (int64_t)2 * w + 2 + h + h / 2; };
      while (w0 < 12 && (d.ext[0] + Wof(w0) - 1) / Wof(w0) + 1 > slots) ++w0;
    } else if (s3_class && p->hd == 1) {
      h = 2; w0 = 7;  // streaming kernel: Table 4's h = 2; two CTAs per SM
    } else {
      // the tile-size model (tilemodel.cpp: Sec. 3.7's load-to-compute ratio with the
      // instruction-cache and CTA-count terms) over the compiled variants of the fast kernel
      // that will run, or over modest hexagons for the generic executor
      const bool unit = p->d0.n == 1 && p->d0.d == 1 && p->d1.n == 1 && p->d1.d == 1 && p->hd == 0;
      int fam = FAMILY_GENERIC;
      if (flags == STENCIL_EXEC_AUTO && unit && d.kind != STENCIL_LINEAR)
        fam = d.dims == 2 ? FAMILY_FAST2D : FAMILY_FAST3D;
      if (!tile_select(d, p->hd, p->d0, p->d1, fam, &h, &w0) &&
          !tile_select(d, p->hd, p->d0, p->d1, FAMILY_GENERIC, &h, &w0)) {
        h = 2;
        w0 = 7;  // Table 4 setup
      }
    }
  }
  if (h < 0 || w0 < 0) return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: negative tile parameter");
  if (2 * h + 2 > kMaxLevels)
    return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: 2h+2 exceeds the kernels' level limit (64)");
  const int64_t wb = w0_bound(p->d0, p->d1, h);
  if (w0 < wb)
    return fail(STENCIL_E_INFEASIBLE_TILE,
                "stencil_plan: w0 violates eq. (1): need w0 >= " + std::to_string(wb));
  p->h = h;
  p->w0 = w0;
  p->F0 = (int)floor_rat_mul(p->d0, h);
  p->F1 = (int)floor_rat_mul(p->d1, h);
  p->H = 2 * h + 2;
  p->W = 2 * w0 + 2 + p->F0 + p->F1;
  p->c = p->F1 - p->F0;
  p->lo.assign(p->H, 0);
  p->hi.assign(p->H, -1);
  for (int a = 0; a < p->H; ++a) {
    int lo = -1, hi = -2;
    for (int b = 0; b < p->W; ++b) {
      if (in_hexagon(*p, a, b)) {
        if (lo < 0) lo = b;
        else if (b != hi + 1) return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: non-convex hexagon row");
        hi = b;
      }
    }
    if (lo < 0) return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: empty hexagon row");
    p->lo[a] = lo;
    p->hi[a] = hi;
  }
  hexagon_traffic(*p);

  // executor selection
  int ex = EXEC_GENERIC;
  p->variant = -1;
  if (flags == STENCIL_EXEC_NAIVE) {
    ex = EXEC_NAIVE;
  } else if (flags == STENCIL_EXEC_AUTO) {
    if (d.kind == STENCIL_FDTD2D) {
      p->variant = fdtd_variant(dtype, h, w0);
      // the ring is filled by 16-B cp.async: row starts must be 16-B aligned
      if (p->variant >= 0 && p->hd == 0 && (d.ext[1] * (int64_t)d.elem()) % 16 == 0) ex = EXEC_FDTD;
    } else if (d.dims == 2) {
      p->variant = fast2d_variant(d.kind, dtype, h, w0, t.w[0]);
      // the kernel's column arithmetic is 32-bit (chunk origins, row bounds): rows of 2^30
      // columns or more take the generic executor
      if (p->variant >= 0 && p->hd == 0 && p->dcls[0] == 1 && p->d0.n == 1 && p->d0.d == 1 &&
          p->d1.n == 1 && p->d1.d == 1 && d.ext[1] < (int64_t(1) << 30) && d.ext[0] < (int64_t(1) << 30))
        ex = EXEC_FAST2D;
    } else if (s3_class && p->hd == 1) {
      p->variant = stream3d_variant(d.kind, dtype, h, w0);
      if (p->variant >= 0 && p->d0.n == 1 && p->d0.d == 1 && p->d1.n == 1 && p->d1.d == 1) ex = EXEC_STREAM3D;
    } else {
      p->variant = fast3d_variant(d.kind, dtype, h, w0, t.w[0]);
      // tuning aid: HEXS_F3_FORCE_VARIANT=<id> picks a compiled variant of the same shape
      if (const char* fv = std::getenv("HEXS_F3_FORCE_VARIANT")) {
        const int id = std::atoi(fv);
        if (id >= 0 && fast3d_variant_matches(id, d.kind, dtype, h, w0)) p->variant = id;
      }
      // TMA tensor maps need 16-B aligned plane/line strides (N2 * elem % 16 == 0)
      // the kernel's hexagon is the unit-slope closed form (compile-time rows per level)
      if (p->variant >= 0 && p->hd == 0 && (d.ext[2] * (int64_t)d.elem()) % 16 == 0 && p->d0.n == 1 &&
          p->d0.d == 1 && p->d1.n == 1 && p->d1.d == 1)
        ex = EXEC_FAST3D;
    }
  } else if (ablation) {
    // Table 4 replay: the 3D radius-1 single-field classes in fp32, hexagons over z, unit skews
    if (d.dims != 3 || !(d.kind == STENCIL_STAR3D7 || d.kind == STENCIL_BOX3D27 || d.kind == STENCIL_GRADIENT3D) ||
        d.dtype != STENCIL_F32 || p->hd != 0 || !(p->d0.n == 1 && p->d0.d == 1 && p->d1.n == 1 && p->d1.d == 1) ||
        p->dcls[0] != 1 || p->dcls[1] != 1)
      return fail(STENCIL_E_UNSUPPORTED,
                  "stencil_plan: the Table 4 executors take 3D radius-1 star3d7/box3d27/gradient3d fp32, hex_dim 0");
    if (!((t.w[0] == 0 && t.w[1] == 0) || (t.w[0] == 10 && t.w[1] == 32)))
      return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: the Table 4 executors use w = {10, 32} (PAPER.md:998-1000)");
    ex = EXEC_ABLATION;
    p->variant = flags - STENCIL_EXEC_T4A;
    const int YB = p->H + 11, XB = p->H + 33, XP = p->variant == 4 ? 64 : XB;
    if (XB > 64 || 2.0 * (p->W + 2) * YB * XP * 4 > 227.0 * 1024)
      return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: the Table 4 copy-in box exceeds shared memory");
  } else if (flags != STENCIL_EXEC_GENERIC) {
    return fail(STENCIL_E_INVALID, "stencil_plan: unknown tile.flags");
  }
  p->executor = ex;

  // classical widths
  for (int q = 0; q < p->ncls; ++q) {
    int wq = t.w[q];
    if (ex == EXEC_FAST2D) wq = fast2d_chunk_width(p->variant);
    else if (ex == EXEC_ABLATION) wq = q == 0 ? 10 : 32;  // Table 4: w1 = 10, w2 = 32
    else if (ex == EXEC_STREAM3D) wq = q == 0 ? 1 : kStream3DNXPlan;  // z planes streamed; x strips
    else if (ex == EXEC_FAST3D) {
      int wy = 0, wx = 0;
      fast3d_tile(p->variant, &wy, &wx);
      wq = q == 0 ? wy : wx;
    } else if (wq <= 0) {
      if (d.dims == 3) wq = (q == p->ncls - 1) ? 64 : 8;  // wavefront tiles (y 8 x 64)
      else wq = (q == p->ncls - 1) ? 128 : 4;
    }
    if (wq < 1) return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_plan: classical width must be >= 1");
    p->w[q] = wq;
  }

  // The 3D fast kernel moves whole 16-B groups (TMA boxes, vector loads/stores): it skews the
  // contiguous dimension by 4 per level (any integer skew >= delta1_i keeps eq. (14) valid,
  // reading R16), so every tile boundary of every level is 16-B aligned.
  if (ex == EXEC_FAST3D || ex == EXEC_STREAM3D) {
    p->dcls[1] = std::max(p->dcls[1], 4);
    p->ctrans[1] = 0;
  }
  // Table 4 (d)-(f) translate the x tiles (Sec. 4.2.3's offset): (d) so the
  // copy-in box [B2 - H, B2 + 33) of a full launch starts on a 128-B line, (e)/(f) so the 32
  // columns each later tile loads, [B2 + 1, B2 + 33), are one aligned line
  if (ex == EXEC_ABLATION) {
    p->ctrans[0] = 0;
    p->ctrans[1] = p->variant == 3 ? p->H % 32 : (p->variant >= 4 ? 31 : 0);
  }

  // a3: launch table.  Order (T, 0), (T, 1), T ascending.
  int64_t dlo[3], dhi[3];
  for (int q = 0; q < d.dims; ++q) {
    dlo[q] = INT64_MAX;
    dhi[q] = INT64_MIN;
    for (auto& st : d.stmts) {
      dlo[q] = std::min<int64_t>(dlo[q], st.lo[q]);
      dhi[q] = std::max<int64_t>(dhi[q], d.ext[q] + st.hi[q] - 1);
    }
  }
  const int64_t L = p->tau_levels;
  if (ex != EXEC_NAIVE && L > 0) {
    const int64_t Tmax0 = floor_div(L - 1 + h + 1, p->H), Tmax1 = floor_div(L - 1, p->H);
    for (int64_t T = 0; T <= std::max(Tmax0, Tmax1); ++T) {
      for (int ph = 0; ph < 2; ++ph) {
        if ((ph == 0 && T > Tmax0) || (ph == 1 && T > Tmax1)) continue;
        Launch ln{};
        ln.T = T;
        ln.phase = ph;
        ln.tau0 = ph == 0 ? T * p->H - (h + 1) : T * p->H;
        ln.a_lo = (int)std::max<int64_t>(0, -ln.tau0);
        ln.a_hi = (int)std::min<int64_t>(p->H - 1, L - 1 - ln.tau0);
        if (ln.a_lo > ln.a_hi) continue;
        ln.row_off = T * p->c + (ph == 0 ? p->F0 + w0 + 1 : 0) + p->hex_origin;
        int bmin = INT32_MAX, bmax = INT32_MIN;
        for (int a = ln.a_lo; a <= ln.a_hi; ++a) {
          bmin = std::min(bmin, (int)p->lo[a]);
          bmax = std::max(bmax, (int)p->hi[a]);
        }
        const int hd = p->hd;
        ln.S0_lo = ceil_div(dlo[hd] + ln.row_off - bmax, p->W);
        ln.S0_hi = floor_div(dhi[hd] + ln.row_off - bmin, p->W);
        if (ln.S0_lo > ln.S0_hi) continue;
        for (int q = 0; q < 2; ++q) {
          ln.Slo[q] = ln.Shi[q] = 0;
          if (q < p->ncls) {
            const int dq = p->cls[q];
            ln.Slo[q] = floor_div(dlo[dq] - p->ctrans[q] + (int64_t)p->dcls[q] * ln.a_lo, p->w[q]);
            ln.Shi[q] = floor_div(dhi[dq] - p->ctrans[q] + (int64_t)p->dcls[q] * ln.a_hi, p->w[q]);
          }
        }
        p->launches.push_back(ln);
      }
    }
  }

  // workspace: the second ping-pong buffer, 256-B granular
  p->ws_bytes = 0;
  if (d.pingpong && T_steps > 0) p->ws_bytes = ((size_t)d.points() * d.elem() + 255) / 256 * 256;
  // 3D generic executor: classical tiles run as a dependence wavefront; per-tile completion
  // flags and a work counter follow the ping-pong buffer in the workspace.
  p->wavefront = ((ex == EXEC_GENERIC || ex == EXEC_FAST3D || ex == EXEC_ABLATION) && d.dims == 3 && p->ncls == 2);
  if (p->wavefront && !p->launches.empty()) {
    // every launch owns its flags and work counter, so one memset per stencil_run resets
    // them all (no reset between the launches of a run)
    int64_t n_items = 0, idx = 0;
    for (Launch& l : p->launches) {
      l.flag_first = n_items;
      l.counter_idx = idx++;
      // (the Table 4 kernel keeps one progress counter per (hexagon, y tile) row)
      n_items += (l.S0_hi - l.S0_lo + 1) * (l.Shi[0] - l.Slo[0] + 1) *
                 (ex == EXEC_ABLATION ? 1 : (l.Shi[1] - l.Slo[1] + 1));
    }
    p->flag_off = p->ws_bytes;
    p->counter_off = p->flag_off + ((size_t)n_items * sizeof(int) + 255) / 256 * 256;
    // flags + ticket counters + per-launch completed-tile counters (3D chained launches)
    p->flag_bytes = p->counter_off - p->flag_off + ((size_t)idx * 16 + 255) / 256 * 256;
    p->n_counters = idx;
    p->ws_bytes = p->flag_off + p->flag_bytes;
  }
  // streaming 3D kernel: per launch a progress counter per (hexagon, strip) CTA plus a ticket
  // (zeroed together by one memset per run), and the carry scratch ring shared by the
  // launches (they run one after the other on the stream)
  if (ex == EXEC_STREAM3D && !p->launches.empty()) {
    p->s3_nstr = (int)((d.ext[2] - 1 + 4 * (p->H - 1)) / kStream3DNXPlan + 1);
    int64_t ctr = 0, max_items = 0;
    for (Launch& l : p->launches) {
      const int64_t items = (l.S0_hi - l.S0_lo + 1) * p->s3_nstr;
      if (items > INT32_MAX / 2) return fail(STENCIL_E_UNSUPPORTED, "stencil_plan: too many tiles per launch");
      l.s3_ctr_first = ctr;
      ctr += items + 1;  // counters, then the ticket
      max_items = std::max(max_items, items);
    }
    p->s3_ctr_off = p->ws_bytes;
    p->s3_ctr_bytes = ((size_t)ctr * sizeof(int) + 255) / 256 * 256;
    p->s3_scratch_off = p->s3_ctr_off + p->s3_ctr_bytes;
    const size_t cblk = (size_t)stream3d_carry_block(p->variant) * sizeof(float);
    p->ws_bytes = p->s3_scratch_off + ((size_t)max_items * kStream3DRSPlan * cblk + 255) / 256 * 256;
  }
  *out = guard.release();
  return STENCIL_OK;
}

}  // namespace hexs

using namespace hexs;

static Plan* as_plan(stencil_plan_t h) {
  Plan* p = reinterpret_cast<Plan*>(h);
  return (p && p->magic == kPlanMagic) ? p : nullptr;
}

extern "C" {

stencil_status stencil_plan(stencil_plan_t* out, stencil_desc_t desc, int64_t T_steps,
                            const stencil_tile_t* tile) {
  clear_error();
  if (!out) return fail(STENCIL_E_INVALID, "stencil_plan: out is NULL");
  *out = nullptr;
  Desc* d = reinterpret_cast<Desc*>(desc);
  if (!d || d->magic != kDescMagic) return fail(STENCIL_E_INVALID, "stencil_plan: bad descriptor");
  Plan* p = nullptr;
  stencil_status s = build_plan(*d, T_steps, tile, &p);
  if (s != STENCIL_OK) return s;
  *out = reinterpret_cast<stencil_plan_t>(p);
  return STENCIL_OK;
}

stencil_status stencil_plan_workspace_size(stencil_plan_t plan, size_t* bytes) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !bytes) return fail(STENCIL_E_INVALID, "stencil_plan_workspace_size: bad arguments");
  *bytes = p->ws_bytes;
  return STENCIL_OK;
}

stencil_status stencil_plan_set_workspace(stencil_plan_t plan, void* dev_ptr, size_t bytes) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p) return fail(STENCIL_E_INVALID, "stencil_plan_set_workspace: bad plan");
  if (bytes < p->ws_bytes) return fail(STENCIL_E_OOM, "stencil_plan_set_workspace: workspace too small");
  if (p->ws_bytes && !dev_ptr) return fail(STENCIL_E_INVALID, "stencil_plan_set_workspace: NULL workspace");
  if (reinterpret_cast<uintptr_t>(dev_ptr) % 256 != 0)
    return fail(STENCIL_E_INVALID, "stencil_plan_set_workspace: workspace must be 256-B aligned");
  p->ws = dev_ptr;
  p->ws_size = bytes;
  if (p->dist) return dist_set_workspace(*p, dev_ptr, bytes);  // shared by the block plans
  return STENCIL_OK;
}

stencil_status stencil_plan_info(stencil_plan_t plan, stencil_plan_info_t* info) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !info) return fail(STENCIL_E_INVALID, "stencil_plan_info: bad arguments");
  if (p->dist) {  // a distributed plan describes its primary local block plan
    stencil_plan_t bp = nullptr;
    stencil_status st = stencil_dist_block_plan(plan, 0, &bp);
    if (st != STENCIL_OK) return st;
    st = stencil_plan_info(bp, info);
    if (st != STENCIL_OK) return st;
    dist_fill_info(*p, *info);
    return STENCIL_OK;
  }
  stencil_plan_info_t& o = *info;
  o = stencil_plan_info_t{};
  const Desc& d = p->desc;
  o.dims = d.dims;
  o.kind = d.kind;
  o.dtype = d.dtype;
  o.n_fields = d.nfields;
  o.statements = (int32_t)d.stmts.size();
  o.hex_dim = p->hd;
  o.delta0_num = (int32_t)p->d0.n;
  o.delta0_den = (int32_t)p->d0.d;
  o.delta1_num = (int32_t)p->d1.n;
  o.delta1_den = (int32_t)p->d1.d;
  for (int q = 0; q < 3; ++q) o.delta_cls[q] = q < p->ncls ? p->dcls[q] : 0;
  for (int q = 0; q < 3; ++q) o.trans_cls[q] = q < p->ncls ? p->ctrans[q] : 0;
  o.h = p->h;
  o.w0 = p->w0;
  for (int q = 0; q < 3; ++q) o.w[q] = q < p->ncls ? p->w[q] : 0;
  o.H = p->H;
  o.W = p->W;
  o.F0 = p->F0;
  o.F1 = p->F1;
  o.executor = p->executor == EXEC_NAIVE       ? STENCIL_EXEC_NAIVE
               : p->executor == EXEC_GENERIC   ? STENCIL_EXEC_GENERIC
               : p->executor == EXEC_ABLATION ? STENCIL_EXEC_T4A + p->variant
                                               : STENCIL_EXEC_AUTO;
  o.fast_kernel = (p->executor == EXEC_FAST2D || p->executor == EXEC_FDTD || p->executor == EXEC_FAST3D ||
                   p->executor == EXEC_STREAM3D);
  o.kernel = p->executor == EXEC_FAST2D ? STENCIL_KERNEL_FAST2D
           : p->executor == EXEC_FDTD ? STENCIL_KERNEL_FDTD
           : p->executor == EXEC_FAST3D ? STENCIL_KERNEL_FAST3D
           : p->executor == EXEC_STREAM3D ? STENCIL_KERNEL_STREAM3D
           : p->executor == EXEC_ABLATION ? STENCIL_KERNEL_ABLATION
           : p->executor == EXEC_NAIVE ? STENCIL_KERNEL_NAIVE : STENCIL_KERNEL_GENERIC;
  o.n_launches = p->executor == EXEC_NAIVE ? p->tau_levels : (int64_t)p->launches.size();
  o.T_steps = p->T_steps;
  o.tau_levels = p->tau_levels;
  int64_t interior = 1;
  if (d.kind == STENCIL_FDTD2D) interior = d.ext[0] * d.ext[1];
  else
    for (int q = 0; q < d.dims; ++q) interior *= (d.ext[q] - 2 * d.radius);
  o.updates = interior * p->T_steps;
  o.tile_points = p->tile_points;
  o.tile_in = p->tile_in;
  o.tile_out = p->tile_out;
  o.workspace_bytes = p->ws_bytes;
  return STENCIL_OK;
}

stencil_status stencil_plan_launches(stencil_plan_t plan, stencil_launch_t* out, int64_t cap,
                                     int64_t* n) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !n) return fail(STENCIL_E_INVALID, "stencil_plan_launches: bad arguments");
  *n = (int64_t)p->launches.size();
  if (!out) return STENCIL_OK;
  if (cap < *n) return fail(STENCIL_E_INVALID, "stencil_plan_launches: capacity too small");
  for (size_t i = 0; i < p->launches.size(); ++i) {
    const Launch& l = p->launches[i];
    out[i] = stencil_launch_t{l.T, l.phase, l.a_lo, l.a_hi, l.tau0, l.S0_lo, l.S0_hi, l.row_off};
  }
  return STENCIL_OK;
}

stencil_status stencil_plan_hexagon(stencil_plan_t plan, int32_t* lo, int32_t* hi, int32_t cap) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !lo || !hi || cap < p->H) return fail(STENCIL_E_INVALID, "stencil_plan_hexagon: bad arguments");
  for (int a = 0; a < p->H; ++a) {
    lo[a] = p->lo[a];
    hi[a] = p->hi[a];
  }
  return STENCIL_OK;
}

stencil_status stencil_plan_schedule_of(stencil_plan_t plan, int64_t tau, const int64_t* s,
                                        int64_t* sched) {
  clear_error();
  Plan* p = as_plan(plan);
  if (!p || !s || !sched) return fail(STENCIL_E_INVALID, "stencil_plan_schedule_of: bad arguments");
  if (!schedule_of(*p, tau, s, sched))
    return fail(STENCIL_E_INVALID, "stencil_plan_schedule_of: point not covered (schedule bug)");
  return STENCIL_OK;
}

}  // extern "C"

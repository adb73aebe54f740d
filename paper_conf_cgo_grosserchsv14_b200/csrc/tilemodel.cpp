// tilemodel.cpp -- automatic tile-size selection (a2): the load-to-compute model of Sec. 3.7
// extended with the two B200 terms the measured tile sweeps show
// (profiles/round1/tile_sweep_*.txt).
//
//   paper:  tile sizes are chosen "to minimize the load-to-compute ratio" -- for a full hexagon
//           per classical column, points P = (h+1)(2w0+2+(delta0+delta1)h)
//           against the values it must load (In) and store (Out); here counted exactly by
//           enumerating the hexagon of eqs. (6)-(13) for any slopes, so
//               B(h, w0) = word * (In + Out) / P          [HBM bytes per update]
//           and the HBM-bound rate is BW / B;
//   B200:   (1) on-chip capacity: the fast kernels unroll every level and row of the hexagon
//           (constraint-based unrolling), so their code grows with P; once a
//           body outgrows the instruction cache the SM starves for instructions (ncu stall
//           "no_instruction") -- factor min(1, C / S)^3, S = P * (4 * flops + 6|10) * 16 bytes,
//           C = 39 000 B (2D register-wavefront kernel; 44 000 before the round-2 select-free
//           body made (2,7) beat (3,7) for star2d5) / 58 000 B (3D tile-wavefront kernel),
//           fitted to the sweeps;
//           (2) CTA count: a launch of n hexagon CTAs on `slots` resident slots runs
//           ceil(n / slots) waves -- factor n / (waves * slots) (grid quantisation).
//   rate = BW / B * code * waves.  Over the compiled fast-kernel variants of a class it picks the
//   measured best tile of every class on B200 (tests/test_tilemodel.py); the generic executor
//   (rolled loops, no code term) takes the lowest B among modest hexagons.
#include <algorithm>
#include <cmath>
#include <set>

#include <cuda_runtime.h>

#include "internal.h"

namespace hexs {

namespace {

int sm_count() {
  int dev = 0, sms = 0;
  if (cudaGetDevice(&dev) == cudaSuccess && cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) == cudaSuccess &&
      sms > 0)
    return sms;
  cudaGetLastError();
  return 148;
}

int flops_of(int kind) {  // FP operations per point (Table 3), sqrt/div counted as ~15 each
  switch (kind) {
    case STENCIL_JACOBI2D5: return 5;
    case STENCIL_STAR2D5: return 6;
    case STENCIL_BOX2D9: return 9;
    case STENCIL_STAR3D7: return 8;
    case STENCIL_BOX3D27: return 27;
    case STENCIL_GRADIENT2D: return 40;
    case STENCIL_GRADIENT3D: return 46;
    default: return 8;
  }
}

int64_t floor_mul(const Rat& r, int64_t h) { return floor_div(r.n * h, r.d); }

}  // namespace

bool tile_eval(const Desc& d, int hd, const Rat& d0, const Rat& d1, int h, int w0, int family, TileEval* out) {
  if (h < 0 || w0 < 0 || 2 * h + 2 > kMaxLevels) return false;
  // the hexagon of eqs. (6)-(13) for these parameters (same arithmetic as the planner)
  const int64_t F0 = floor_mul(d0, h), F1 = floor_mul(d1, h);
  const int64_t H = 2 * (int64_t)h + 2, W = 2 * (int64_t)w0 + 2 + F0 + F1;
  const int64_t n0 = d0.n, q0 = d0.d, n1 = d1.n, q1 = d1.d;
  auto inside = [&](int64_t a, int64_t b) {
    if (a < 0 || a > 2 * h + 1) return false;
    if (n0 * a - b * q0 > (2 * h + 1) * n0 - F0 * q0) return false;
    if (n1 * a + b * q1 > (2 * h + 1) * n1 + (F0 + w0) * q1) return false;
    if (n1 * a + b * q1 < h * n1 - (q1 - 1)) return false;
    if (n0 * a - b * q0 < h * n0 - (F0 + w0 + F1) * q0 - (q0 - 1)) return false;
    return true;
  };
  std::set<int> offs;
  for (auto& st : d.stmts)
    for (auto& ac : st.reads) offs.insert(ac.off[hd]);
  std::set<std::pair<int64_t, int64_t>> ins;
  int64_t P = 0, O = 0;
  for (int64_t a = 0; a < H; ++a)
    for (int64_t b = 0; b < W; ++b) {
      if (!inside(a, b)) continue;
      ++P;
      bool is_out = false;
      for (int o : offs) {
        if (!inside(a - 1, b + o)) ins.insert({a - 1, b + o});
        if (!inside(a + 1, b - o)) is_out = true;
      }
      O += is_out;
    }
  if (P == 0) return false;
  TileEval e{};
  e.h = h;
  e.w0 = w0;
  e.points = P;
  e.in = (int64_t)ins.size();
  e.out = O;
  e.bytes_per_update = (double)d.elem() * (double)(e.in + O) / (double)P;
  const double bw = 6.54e12;  // measured copy bandwidth (MEASURED_PEAKS.json); a constant for ranking
  // unrolled body: per hexagon point and column, 4 points per thread of flops each plus the
  // per-row data movement (shuffles, shared loads, stores): 6 (2D) / 10 (3D) instructions of 16 B
  const double per_row = family == FAMILY_FAST2D ? 4.0 * flops_of(d.kind) + 6.0 : 4.0 * flops_of(d.kind) + 10.0;
  e.body_bytes = family == FAMILY_GENERIC ? 0.0 : (double)P * per_row * 16.0;
  const double cap = family == FAMILY_FAST2D ? 39000.0 : 58000.0;
  e.code_eff = family == FAMILY_GENERIC ? 1.0 : std::pow(std::min(1.0, cap / e.body_bytes), 3.0);
  // CTA count: one CTA per hexagon of a launch (2D fast and generic kernels: 3 resident per
  // SM); the 3D kernels are persistent over (hexagon, classical tile) items
  e.ctas = (d.ext[hd] + W - 1) / W;
  e.slots = (int64_t)sm_count() * 3;
  if (family == FAMILY_FAST3D) {
    e.wave_eff = 1.0;
  } else {
    const int64_t waves = (e.ctas + e.slots - 1) / e.slots;
    e.wave_eff = (double)e.ctas / (double)(waves * e.slots);
  }
  e.rate = bw / e.bytes_per_update * e.code_eff * e.wave_eff;
  *out = e;
  return true;
}

bool tile_select(const Desc& d, int hd, const Rat& d0, const Rat& d1, int family, int* h, int* w0) {
  TileEval best{};
  bool have = false;
  auto consider = [&](int hh, int ww) {
    TileEval e;
    if (!tile_eval(d, hd, d0, d1, hh, ww, family, &e)) return;
    if (!have || e.rate > best.rate * (1.0 + 1e-9)) {
      best = e;
      have = true;
    }
  };
  if (family == FAMILY_FAST2D) {
    for (int v = 0; v < fast2d_variant_count(); ++v) {
      int k, dt, hh, ww;
      if (fast2d_variant_info(v, &k, &dt, &hh, &ww) && k == d.kind && dt == d.dtype) consider(hh, ww);
    }
  } else if (family == FAMILY_FAST3D) {
    for (int v = 0; v < fast3d_variant_count(); ++v) {
      int k, dt, hh, ww;
      if (fast3d_variant_info(v, &k, &dt, &hh, &ww) && k == d.kind && dt == d.dtype) consider(hh, ww);
    }
  } else {
    // generic executor: modest hexagons (at most 8 levels, w0 within 12 of eq. (1)'s bound)
    // with enough hexagons per launch to occupy the SMs when the grid allows it
    for (int hh = 1; hh <= 3; ++hh) {
      // eq. (1): w0 >= max(d0 + {d0 h}, d1 + {d1 h}) - 1
      auto term = [&](const Rat& r) {
        const int64_t num = r.n + (r.n * hh - floor_mul(r, hh) * r.d) - r.d;
        return ceil_div(num, r.d);
      };
      const int wb = (int)std::max<int64_t>(0, std::max(term(d0), term(d1)));
      for (int ww = wb; ww <= wb + 12; ++ww) {
        TileEval e;
        if (!tile_eval(d, hd, d0, d1, hh, ww, family, &e)) continue;
        if (e.ctas < sm_count() && ww > wb) continue;  // keep the hexagon count up on small grids
        consider(hh, ww);
      }
    }
  }
  if (!have) return false;
  *h = best.h;
  *w0 = best.w0;
  return true;
}

}  // namespace hexs

using namespace hexs;

extern "C" stencil_status stencil_tile_model(stencil_desc_t desc, int h, int w0, int hex_dim, int family,
                                             stencil_tile_eval_t* out) {
  clear_error();
  Desc* d = reinterpret_cast<Desc*>(desc);
  if (!d || d->magic != kDescMagic || !out) return fail(STENCIL_E_INVALID, "stencil_tile_model: bad arguments");
  if (hex_dim < 0 || hex_dim >= d->dims - 1) return fail(STENCIL_E_INVALID, "stencil_tile_model: bad hex_dim");
  // cone slopes along hex_dim from the dependence distances (as the planner computes them)
  Rat s0 = make_rat(0, 1), s1 = make_rat(0, 1);
  for (auto& v : dependence_distances(*d)) {
    Rat fwd = make_rat(v[1 + hex_dim], v[0]), bwd = make_rat(-v[1 + hex_dim], v[0]);
    if (rat_less(s0, fwd)) s0 = fwd;
    if (rat_less(s1, bwd)) s1 = bwd;
  }
  TileEval e;
  if (!tile_eval(*d, hex_dim, s0, s1, h, w0, family, &e))
    return fail(STENCIL_E_INFEASIBLE_TILE, "stencil_tile_model: not a valid hexagon");
  stencil_tile_eval_t o{};
  o.h = e.h;
  o.w0 = e.w0;
  o.points = e.points;
  o.in = e.in;
  o.out = e.out;
  o.bytes_per_update = e.bytes_per_update;
  o.body_bytes = e.body_bytes;
  o.code_eff = e.code_eff;
  o.ctas = e.ctas;
  o.slots = e.slots;
  o.wave_eff = e.wave_eff;
  o.rate = e.rate;
  int sh = 0, sw = 0;
  o.selected = tile_select(*d, hex_dim, s0, s1, family, &sh, &sw) && sh == h && sw == w0;
  *out = o;
  return STENCIL_OK;
}

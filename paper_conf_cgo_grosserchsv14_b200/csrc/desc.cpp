// desc.cpp -- stencil descriptors, the statement model and dependence analysis (a1).
//
// Sec. 3.2: the input is an outer time loop around k >= 1 perfect
// nests without carried dependences; the canonical schedule is L_i[t, s] -> [k*t+i, s].
// Sec. 3.1: dependences follow from the iteration domains, the
// access relations and the original order.  For the fixed statement shapes of this
// library the memory-based distance set is finite and is enumerated in closed form here
// (the brute-force simulation in oracle/schedule.py pins it in the tests).
#include <algorithm>
#include <cstdlib>
#include <cstring>
#include <new>
#include <set>

#include "internal.h"

namespace hexs {

static thread_local std::string g_err;

stencil_status fail(stencil_status s, const std::string& msg) {
  g_err = msg;
  return s;
}
void clear_error() { g_err.clear(); }

int64_t floor_div(int64_t a, int64_t b) {
  int64_t q = a / b, r = a % b;
  return (r != 0 && ((r < 0) != (b < 0))) ? q - 1 : q;
}
int64_t ceil_div(int64_t a, int64_t b) { return -floor_div(-a, b); }

static int64_t gcd64(int64_t a, int64_t b) {
  if (a < 0) a = -a;
  if (b < 0) b = -b;
  while (b) {
    int64_t t = a % b;
    a = b;
    b = t;
  }
  return a ? a : 1;
}
Rat make_rat(int64_t n, int64_t d) {
  if (d < 0) {
    n = -n;
    d = -d;
  }
  int64_t g = gcd64(n, d);
  return Rat{n / g, d / g};
}
bool rat_less(const Rat& a, const Rat& b) { return a.n * b.d < b.n * a.d; }

// ---------------------------------------------------------------------------------
// Statement models of the classes (access sets of Table 3 / Fig. 1).
// ---------------------------------------------------------------------------------
static int class_dims(int kind) {
  switch (kind) {
    case STENCIL_JACOBI2D5: case STENCIL_STAR2D5: case STENCIL_BOX2D9:
    case STENCIL_FDTD2D: case STENCIL_GRADIENT2D: return 2;
    case STENCIL_STAR3D7: case STENCIL_GRADIENT3D: case STENCIL_BOX3D27: return 3;
    case STENCIL_LINEAR: return -1;  // 2 or 3
    default: return 0;
  }
}

static std::vector<std::vector<int>> class_offsets(int kind) {
  std::vector<std::vector<int>> o;
  switch (kind) {
    case STENCIL_JACOBI2D5: case STENCIL_STAR2D5: case STENCIL_GRADIENT2D:
      o = {{0, 0}, {-1, 0}, {1, 0}, {0, -1}, {0, 1}};
      break;
    case STENCIL_BOX2D9:
      for (int a = -1; a <= 1; ++a)
        for (int b = -1; b <= 1; ++b) o.push_back({a, b});
      break;
    case STENCIL_STAR3D7: case STENCIL_GRADIENT3D:
      o = {{0, 0, 0}, {-1, 0, 0}, {1, 0, 0}, {0, -1, 0}, {0, 1, 0}, {0, 0, -1}, {0, 0, 1}};
      break;
    case STENCIL_BOX3D27:
      for (int a = -1; a <= 1; ++a)
        for (int b = -1; b <= 1; ++b)
          for (int c = -1; c <= 1; ++c) o.push_back({a, b, c});
      break;
    default:
      break;
  }
  return o;
}

static void default_coefficients(int kind, double* c, int* n) {
  switch (kind) {
    case STENCIL_JACOBI2D5: c[0] = 0.2; *n = 1; break;           // Fig. 1
    case STENCIL_STAR2D5: c[0] = 0.5; c[1] = 0.125; *n = 2; break;
    case STENCIL_BOX2D9: c[0] = 1.0 / 9.0; *n = 1; break;
    case STENCIL_FDTD2D: c[0] = 0.5; c[1] = 0.7; *n = 2; break;  // PolyBench fdtd-2d
    case STENCIL_STAR3D7: c[0] = 0.25; c[1] = 0.125; *n = 2; break;
    case STENCIL_GRADIENT3D: c[0] = 1e-2; *n = 1; break;
    case STENCIL_BOX3D27: c[0] = 1.0 / 27.0; *n = 1; break;
    case STENCIL_GRADIENT2D: c[0] = 1e-2; *n = 1; break;
    default: *n = 0;
  }
}

static void build_statements(Desc& d) {
  d.stmts.clear();
  if (d.kind == STENCIL_FDTD2D) {
    // fields: 0 = ex, 1 = ey, 2 = hz.  Order within a step: ey, ex, hz (tau = 3t + i).
    d.nfields = 3;
    d.pingpong = false;
    Stmt ey{1, {{1, {0, 0, 0}}, {2, {0, 0, 0}}, {2, {-1, 0, 0}}}, {1, 0, 0}, {0, 0, 0}};
    Stmt ex{0, {{0, {0, 0, 0}}, {2, {0, 0, 0}}, {2, {0, -1, 0}}}, {0, 1, 0}, {0, 0, 0}};
    Stmt hz{2,
            {{2, {0, 0, 0}}, {0, {0, 1, 0}}, {0, {0, 0, 0}}, {1, {1, 0, 0}}, {1, {0, 0, 0}}},
            {0, 0, 0},
            {-1, -1, 0}};
    d.stmts = {ey, ex, hz};
    return;
  }
  d.nfields = 1;
  d.pingpong = true;
  Stmt s;
  s.write = 0;
  std::vector<std::vector<int>> offs = class_offsets(d.kind);
  if (d.kind == STENCIL_LINEAR) {
    offs.clear();
    for (size_t k = 0; k * d.dims < d.loff.size(); ++k)
      offs.push_back(std::vector<int>(d.loff.begin() + k * d.dims, d.loff.begin() + (k + 1) * d.dims));
  }
  for (auto& o : offs) {
    Access a{0, {0, 0, 0}};
    for (int k = 0; k < d.dims; ++k) a.off[k] = o[k];
    s.reads.push_back(a);
  }
  for (int k = 0; k < 3; ++k) {
    s.lo[k] = k < d.dims ? d.radius : 0;
    s.hi[k] = k < d.dims ? -d.radius : 0;
  }
  d.stmts = {s};
}

// Memory-based distance vectors of the canonical schedule.
//   Ping-pong (Fig. 1): instance (t,s) reads A[t%2][s+o] and writes A[(t+1)%2][s]:
//     RAW (1, -o), WAR (1, +o), WAW (2, 0).
//   In place, k statements, tau = k*t + i: for a read of field f at offset o by statement
//   R and the writer W of f, with D(x) = x mod k (0 -> k):
//     RAW W->R: (D(iR - iW), -o);  WAR R->W: (D(iW - iR), +o);  WAW W->W: (k, 0).
std::vector<std::vector<int64_t>> dependence_distances(const Desc& d) {
  std::set<std::vector<int64_t>> out;
  const int k = (int)d.stmts.size();
  auto vec = [&](int64_t dt, const int* off, int sign) {
    std::vector<int64_t> v(1 + d.dims);
    v[0] = dt;
    for (int q = 0; q < d.dims; ++q) v[1 + q] = sign * off[q];
    return v;
  };
  const int zero[3] = {0, 0, 0};
  if (d.pingpong) {
    for (auto& a : d.stmts[0].reads) {
      out.insert(vec(1, a.off, -1));
      out.insert(vec(1, a.off, +1));
    }
    out.insert(vec(2, zero, 1));
  } else {
    auto D = [&](int x) {
      int m = ((x % k) + k) % k;
      return m == 0 ? k : m;
    };
    for (int iR = 0; iR < k; ++iR) {
      for (auto& a : d.stmts[iR].reads) {
        for (int iW = 0; iW < k; ++iW) {
          if (d.stmts[iW].write != a.field) continue;
          out.insert(vec(D(iR - iW), a.off, -1));
          out.insert(vec(D(iW - iR), a.off, +1));
        }
      }
    }
    for (int iW = 0; iW < k; ++iW) out.insert(vec(k, zero, 1));
  }
  return std::vector<std::vector<int64_t>>(out.begin(), out.end());
}

}  // namespace hexs

using namespace hexs;

extern "C" {

int stencil_abi_version(void) { return STENCIL_ABI_VERSION; }

const char* stencil_last_error(void) { return hexs::g_err.c_str(); }

stencil_status stencil_desc_create(stencil_desc_t* out, int dims, const int64_t* extents,
                                   stencil_kind kind, int radius, const int32_t* offsets,
                                   int n_offsets, const double* coefficients,
                                   int n_coefficients, stencil_dtype dtype) {
  clear_error();
  if (!out) return fail(STENCIL_E_INVALID, "stencil_desc_create: out is NULL");
  *out = nullptr;
  const int cd = class_dims(kind);
  if (cd == 0) return fail(STENCIL_E_INVALID, "stencil_desc_create: unknown stencil kind");
  if (cd > 0 ? dims != cd : (dims != 2 && dims != 3))
    return fail(STENCIL_E_INVALID, "stencil_desc_create: dims does not match the class");
  if (!extents) return fail(STENCIL_E_INVALID, "stencil_desc_create: extents is NULL");
  if (kind == STENCIL_LINEAR) {
    if (!offsets || !coefficients || n_offsets < 1 || n_offsets > 64 || n_coefficients != n_offsets)
      return fail(STENCIL_E_INVALID, "stencil_desc_create: LINEAR needs 1..64 offsets and one coefficient each");
    int R = 0;
    for (int q = 0; q < n_offsets * dims; ++q) R = std::max(R, std::abs((int)offsets[q]));
    if (radius != R)
      return fail(STENCIL_E_INVALID, "stencil_desc_create: radius must equal max |offset| of the access set");
    if (R < 1 || R > 8) return fail(STENCIL_E_UNSUPPORTED, "stencil_desc_create: LINEAR radius must be in [1, 8]");
  } else if (radius != 1) {
    return fail(STENCIL_E_UNSUPPORTED, "stencil_desc_create: the fixed classes have radius 1");
  }
  if (dtype != STENCIL_F32 && dtype != STENCIL_F64) return fail(STENCIL_E_INVALID, "stencil_desc_create: bad dtype");
  for (int q = 0; q < dims; ++q)
    if (extents[q] < 2 * radius + 1 || extents[q] > (int64_t(1) << 31))
      return fail(STENCIL_E_INVALID, "stencil_desc_create: every extent must be in [2r+1, 2^31]");
  Desc* d = new (std::nothrow) Desc();
  if (!d) return fail(STENCIL_E_OOM, "stencil_desc_create: out of host memory");
  d->dims = dims;
  for (int q = 0; q < 3; ++q) d->ext[q] = q < dims ? extents[q] : 1;
  d->kind = kind;
  d->radius = radius;
  d->dtype = dtype;
  int nd = 0;
  default_coefficients(kind, d->coef, &nd);
  d->ncoef = nd;
  if (kind == STENCIL_LINEAR) {
    d->loff.assign(offsets, offsets + (size_t)n_offsets * dims);
    d->lcoef.assign(coefficients, coefficients + n_offsets);
    build_statements(*d);
    *out = reinterpret_cast<stencil_desc_t>(d);
    return STENCIL_OK;
  }
  if (coefficients) {
    if (n_coefficients != nd) {
      delete d;
      return fail(STENCIL_E_INVALID, "stencil_desc_create: wrong number of coefficients for the class");
    }
    for (int q = 0; q < nd; ++q) d->coef[q] = coefficients[q];
  }
  if (offsets) {
    if (kind == STENCIL_FDTD2D) {
      delete d;
      return fail(STENCIL_E_INVALID, "stencil_desc_create: FDTD2D takes no offsets (three fixed statements)");
    }
    std::set<std::vector<int>> want, got;
    for (auto& o : class_offsets(kind)) want.insert(o);
    for (int q = 0; q < n_offsets; ++q) {
      std::vector<int> o(dims);
      for (int r = 0; r < dims; ++r) o[r] = offsets[q * dims + r];
      got.insert(o);
    }
    if (want != got || (int)want.size() != n_offsets) {
      delete d;
      return fail(STENCIL_E_INVALID, "stencil_desc_create: offsets do not match the class's access set");
    }
  }
  build_statements(*d);
  *out = reinterpret_cast<stencil_desc_t>(d);
  return STENCIL_OK;
}

stencil_status stencil_desc_deps(stencil_desc_t desc, int32_t* dist, int cap, int* n) {
  clear_error();
  Desc* d = reinterpret_cast<Desc*>(desc);
  if (!d || d->magic != kDescMagic || !n) return fail(STENCIL_E_INVALID, "stencil_desc_deps: bad handle");
  auto v = dependence_distances(*d);
  *n = (int)v.size();
  if (dist) {
    if (cap < (int)v.size()) return fail(STENCIL_E_INVALID, "stencil_desc_deps: capacity too small");
    for (size_t i = 0; i < v.size(); ++i)
      for (int q = 0; q <= d->dims; ++q) dist[i * (d->dims + 1) + q] = (int32_t)v[i][q];
  }
  return STENCIL_OK;
}

stencil_status stencil_destroy(void* handle) {
  clear_error();
  if (!handle) return STENCIL_OK;
  uint32_t magic;
  std::memcpy(&magic, handle, sizeof(magic));
  if (magic == kDescMagic) {
    Desc* d = reinterpret_cast<Desc*>(handle);
    d->magic = 0;
    delete d;
    return STENCIL_OK;
  }
  if (magic == kPlanMagic) {
    Plan* p = reinterpret_cast<Plan*>(handle);
    p->magic = 0;
    delete p;
    return STENCIL_OK;
  }
  return fail(STENCIL_E_INVALID, "stencil_destroy: not a stencil handle");
}

}  // extern "C"

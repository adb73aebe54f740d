"""Small runs of every kernel family through the C ABI, for compute-sanitizer
(memcheck / racecheck / synccheck / initcheck):

    compute-sanitizer --tool racecheck python tools/sanitize_cases.py [case ...]

Device memory comes straight from libcudart via ctypes (no torch: keeps the sanitized
process small).  Each case also checks its result against the oracle, so a run that the
tool slows down or perturbs still has to be bit-exact.  Exit code 0 = all cases passed."""
import ctypes
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import oracle  # noqa: E402  (test infrastructure: the checker)
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import _lib  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200._lib import EXEC, KINDS, Tile, check  # noqa: E402

cudart = ctypes.CDLL("libcudart.so.12")
H2D, D2H = 1, 2


def dmalloc(n):
    p = ctypes.c_void_p()
    assert cudart.cudaMalloc(ctypes.byref(p), ctypes.c_size_t(n)) == 0
    return p


def run_case(kind, shape, T, dtype=np.float32, h=0, w0=0, executor="auto", hex_dim=-1):
    L = _lib.lib()
    nf = 3 if kind == "fdtd2d" else 1
    fields = (stencil_inputs.fields(shape, seed=3, n=3, dtype=dtype) if nf == 3
              else [stencil_inputs.uniform(shape, seed=3, dtype=dtype)])
    ext = (ctypes.c_int64 * len(shape))(*shape)
    d = ctypes.c_void_p()
    check(L.stencil_desc_create(ctypes.byref(d), len(shape), ext, KINDS[kind], 1, None, 0, None, 0,
                                1 if dtype == np.float64 else 0))
    t = Tile(h, w0, (ctypes.c_int32 * 3)(0, 0, 0), hex_dim, EXEC[executor])
    p = ctypes.c_void_p()
    check(L.stencil_plan(ctypes.byref(p), d, T, ctypes.byref(t)))
    ws_n = ctypes.c_size_t()
    check(L.stencil_plan_workspace_size(p, ctypes.byref(ws_n)))
    ws = dmalloc(ws_n.value + 256) if ws_n.value else ctypes.c_void_p()
    check(L.stencil_plan_set_workspace(p, ws, ws_n.value))
    nbytes = fields[0].nbytes
    din = [dmalloc(nbytes) for _ in range(nf)]
    dout = [dmalloc(nbytes) for _ in range(nf)]
    for a, f in zip(din, fields):
        assert cudart.cudaMemcpy(a, f.ctypes.data_as(ctypes.c_void_p), ctypes.c_size_t(nbytes), H2D) == 0
    ip = (ctypes.c_void_p * nf)(*[a.value for a in din])
    op = (ctypes.c_void_p * nf)(*[a.value for a in dout])
    for _ in range(2):  # eager run, then the captured graph's first replay
        check(L.stencil_run(p, ip, op, T, None))
    assert cudart.cudaDeviceSynchronize() == 0
    got = [np.empty_like(fields[0]) for _ in range(nf)]
    for g, a in zip(got, dout):
        assert cudart.cudaMemcpy(g.ctypes.data_as(ctypes.c_void_p), a, ctypes.c_size_t(nbytes), D2H) == 0
    exp = oracle.fdtd(*fields, T) if nf == 3 else [oracle.run(kind, fields[0], T)]
    ok = all(np.array_equal(a, b) for a, b in zip(got, exp))
    for a in din + dout + ([ws] if ws.value else []):
        cudart.cudaFree(a)
    L.stencil_destroy(p)
    L.stencil_destroy(d)
    return ok


CASES = {
    "fast2d": ("star2d5", (70, 1030), 19, np.float32, 3, 7),        # aligned rows, 2 chunks, t-cut tiles
    "fast2d_box": ("box2d9", (45, 531), 11, np.float32, 2, 7),      # unaligned rows
    "fast2d_grad": ("gradient2d", (40, 1024), 9, np.float32, 0, 0),
    "fast2d_f64": ("star2d5", (40, 520), 9, np.float64, 0, 0),
    "stream3d": ("star3d7", (26, 40, 136), 9, np.float32, 0, 0),       # 3 strips, default (2,7)
    "stream3d_grad": ("gradient3d", (22, 36, 68), 7, np.float32, 0, 0),
    "stream3d_h1": ("star3d7", (19, 30, 72), 6, np.float32, 1, 7),
    "fast3d": ("star3d7", (26, 40, 72), 9, np.float32, 0, 0),           # hex_dim 0: tile wavefront
    "fast3d_box": ("box3d27", (20, 34, 64), 7, np.float32, 0, 0),
    "fast3d_f64": ("star3d7", (20, 34, 64), 7, np.float64, 0, 0),
    "fdtd": ("fdtd2d", (60, 136), 9, np.float32, 0, 0),
    "generic3d": ("star3d7", (18, 21, 23), 6, np.float32, 1, 1),
}
# Table 4 replay (kernels/ablation.cu): every memory strategy, 2 x tiles per row and 2 y rows
for _c in "abcdef":
    CASES[f"t4{_c}"] = ("box3d27", (24, 22, 70), 7, np.float32, 0, 0)


def main(argv):
    names = argv or sorted(CASES)
    bad = []
    for n in names:
        kind, shape, T, dt, h, w0 = CASES[n]
        ex = "generic" if n.startswith("generic") else (n if n.startswith("t4") else "auto")
        hd = 0 if n.startswith(("fast3d", "t4")) else (1 if n.startswith("stream3d") else -1)
        ok = run_case(kind, shape, T, dt, h, w0, ex, hd)
        print(f"{n}: {'ok' if ok else 'MISMATCH'}", flush=True)
        if not ok:
            bad.append(n)
    return 1 if bad else 0


if __name__ == "__main__":
    sys.exit(main(sys.argv[1:]))

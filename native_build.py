"""Build the native libraries in-tree (no JIT cache, so the .so files travel to the GPU box).

  * paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil.so -- the product: C++ planner +
    sm_100a CUDA kernels behind include/stencil.h (nvcc -gencode arch=compute_100a,
    code=sm_100a, --fmad=false for bit-exact parity, -lineinfo).
  * oracle/liboracle.so -- the CPU oracle (test infrastructure; built here only so the
    checker exists -- building it is not using it).
"""
from __future__ import annotations

import argparse
import concurrent.futures as cf
import hashlib
import os
import re
import subprocess
import sys

ROOT = os.path.dirname(os.path.abspath(__file__))
PKG = os.path.join(ROOT, "paper_conf_cgo_grosserchsv14_b200")
CSRC = os.path.join(PKG, "csrc")
KDIR = os.path.join(CSRC, "kernels")
OBJ = os.path.join(ROOT, "build", "obj")
LIB = os.path.join(PKG, "lib", "libhexstencil.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")

ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
NVFLAGS = ARCH + ["-O3", "-std=c++17", "-lineinfo", "--fmad=false", "-prec-div=true",
                  "-prec-sqrt=true", "-ftz=false", "-Xcompiler", "-fPIC", "-Xptxas", "-v",
                  "-I", os.path.join(ROOT, "include")]
def _nccl_include():
    """nccl.h of the NCCL the process will load at run time (PyTorch's wheel), else the system's."""
    try:
        import importlib.util

        spec = importlib.util.find_spec("nvidia.nccl")
        if spec and spec.submodule_search_locations:
            inc = os.path.join(list(spec.submodule_search_locations)[0], "include")
            if os.path.exists(os.path.join(inc, "nccl.h")):
                return inc
    except Exception:  # noqa: BLE001
        pass
    return "/usr/include"


CXXFLAGS = ["-O2", "-std=c++17", "-fPIC", "-ffp-contract=off", "-I", os.path.join(ROOT, "include"),
            "-I", "/usr/local/cuda/include", "-I", _nccl_include()]


def _variant_ids(header: str, macro: str):
    txt = open(os.path.join(KDIR, header)).read()
    body = txt.split(f"#define {macro}(X)", 1)[1].split("#define", 1)[0]
    return [int(m) for m in re.findall(r"X\((\d+),", body)]


def _deps_hash(paths):
    h = hashlib.sha1()
    for p in sorted(paths):
        h.update(open(p, "rb").read())
    return h.hexdigest()[:16]


EXTRA3D = []  # extra flags of the 3D kernel objects (debug builds)
EXTRAS3 = []  # extra flags of the streaming 3D kernel objects
EXTRA_ALL = []  # extra flags of the CUDA objects matching EXTRA_ONLY (experiment builds: --variant)
EXTRA_ONLY = [""]


def _units():
    """(source, object, extra flags) for every translation unit."""
    headers = [os.path.join(dp, f) for dp, _, fs in os.walk(CSRC) for f in fs
               if f.endswith((".h", ".cuh"))] + [os.path.join(ROOT, "include", "stencil.h")]
    units = []
    for src in ["desc.cpp", "plan.cpp", "dist.cpp", "tilemodel.cpp"]:
        units.append((os.path.join(CSRC, src), "cxx", []))
    for src in ["run.cu", "kernels/generic.cu", "kernels/registry.cu", "kernels/fdtd.cu",
                "kernels/ablation.cu"]:
        units.append((os.path.join(CSRC, src), "nvcc", []))
    # the halo kernels use NCCL's device API (symmetric-window LSA pointers): nccl_device.h
    units.append((os.path.join(CSRC, "kernels/halo.cu"), "nvcc", ["-I" + _nccl_include()]))
    for vid in _variant_ids("fast2d_variants.h", "HEXS_FAST2D_VARIANTS"):
        units.append((os.path.join(KDIR, "fast2d_inst.cu"), "nvcc", [f"-DHEXS_VARIANT={vid}"]))
    for vid in _variant_ids("fast3d_variants.h", "HEXS_FAST3D_VARIANTS"):
        units.append((os.path.join(KDIR, "hex3d.cu"), "nvcc", [f"-DHEXS_F3_VARIANT={vid}"] + EXTRA3D))
    for vid in _variant_ids("stream3d_variants.h", "HEXS_STREAM3D_VARIANTS"):
        units.append((os.path.join(KDIR, "stream3d.cu"), "nvcc", [f"-DHEXS_S3_VARIANT={vid}"] + EXTRAS3))
    out = []
    if EXTRA_ALL:
        units = [(src, tool, extra + EXTRA_ALL if tool == "nvcc" and EXTRA_ONLY[0] in src else extra)
                 for src, tool, extra in units]
    for src, tool, extra in units:
        key = _deps_hash([src] + headers) + hashlib.sha1(" ".join(extra).encode()).hexdigest()[:8]
        tags = [e.split("=")[-1] for e in extra if "=" in e]
        name = os.path.relpath(src, CSRC).replace("/", "_") + ("_" + "_".join(tags) if tags else "")
        out.append((src, tool, extra, os.path.join(OBJ, f"{name}.{key}.o")))
    return out


def _compile(unit, verbose=False):
    src, tool, extra, obj = unit
    if os.path.exists(obj):
        return obj, ""
    if tool == "cxx":
        cmd = ["g++"] + CXXFLAGS + extra + ["-c", src, "-o", obj]
    else:
        cmd = [NVCC] + NVFLAGS + extra + ["-c", src, "-o", obj]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"compile failed: {' '.join(cmd)}\n{r.stdout}\n{r.stderr}")
    return obj, r.stderr


def build_library(jobs: int = 0, verbose: bool = False, lib: str = None) -> str:
    LIB = lib or globals()["LIB"]
    os.makedirs(OBJ, exist_ok=True)
    os.makedirs(os.path.dirname(LIB), exist_ok=True)
    units = _units()
    jobs = jobs or max(1, os.cpu_count() or 1)
    logs = []
    with cf.ThreadPoolExecutor(jobs) as ex:
        for obj, log in ex.map(lambda u: _compile(u, verbose), units):
            logs.append((obj, log))
    objs = [u[3] for u in units]
    stamp = LIB + ".objs"
    want = "\n".join(objs)
    if not os.path.exists(LIB) or not os.path.exists(stamp) or open(stamp).read() != want:
        cmd = [NVCC] + ARCH + ["-shared", "-o", LIB] + objs + ["-lcudart", "-ldl"]
        subprocess.check_call(cmd)
        open(stamp, "w").write(want)
    if verbose:
        for obj, log in logs:
            if log:
                print(f"== {os.path.basename(obj)}\n{log}")
    return LIB


def build_oracle() -> str:
    sys.path.insert(0, ROOT)
    import oracle  # noqa: E402  (test infrastructure; building the checker is not using it)
    return oracle.build()


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("-j", type=int, default=0)
    ap.add_argument("-v", action="store_true")
    ap.add_argument("--timing", action="store_true",
                    help="also build lib/libhexstencil_tm.so with the 3D kernel's cycle accounting")
    ap.add_argument("--s3trace", action="store_true",
                    help="also build lib/libhexstencil_s3t.so with the streaming 3D kernel's event trace")
    ap.add_argument("--variant", default="",
                    help="build lib/libhexstencil_<VARIANT>.so with the -D flags below instead (experiments; "
                         "load it with HEXS_LIB)")
    ap.add_argument("-D", action="append", default=[], help="macro for the CUDA objects of --variant")
    ap.add_argument("--only", default="", help="apply the -D flags only to sources whose path contains this")
    args = ap.parse_args()
    if args.variant:
        EXTRA_ALL.extend("-D" + d for d in args.D)
        EXTRA_ONLY[0] = args.only
        print(build_library(args.j, args.v, lib=os.path.join(PKG, "lib", f"libhexstencil_{args.variant}.so")))
        return
    print(build_library(args.j, args.v))
    if args.s3trace:
        EXTRAS3.append("-DHEXS_S3_TRACE")
        print(build_library(args.j, args.v, lib=os.path.join(PKG, "lib", "libhexstencil_s3t.so")))
        for tag, flag in ():
            EXTRAS3.append(flag)
            print(build_library(args.j, args.v, lib=os.path.join(PKG, "lib", f"libhexstencil_s3t_{tag}.so")))
            EXTRAS3.remove(flag)
    if args.timing:
        EXTRA3D.append("-DHEXS_F3_TIMING")
        print(build_library(args.j, args.v, lib=os.path.join(PKG, "lib", "libhexstencil_tm.so")))
    print(build_oracle())


if __name__ == "__main__":
    main()

"""Build libaccel.so in-tree with nvcc for sm_100a (B200).

    python -m paper_conf_cgo_margiolaso16_b200.build [--force] [--verbose]

The library is the product: C ABI (include/accel.h) + host runtime + share
solver + device dispatch + tenant kernels.  It statically links the CUDA
runtime, so it does not depend on which libcudart the Python process loaded.
"""
from __future__ import annotations

import glob
import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
INCLUDE = os.path.join(ROOT, "include")
LIB = os.path.join(PKG, "libaccel.so")
LIB_RT = os.path.join(PKG, "libaccel_rt.so")             # same objects, shared CUDA runtime
LIB_INTERCEPT = os.path.join(PKG, "libaccel_intercept.so")
APP = os.path.join(ROOT, "examples", "intercept_app")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
FLAGS = ["-O3", "-lineinfo", "-std=c++17", "-Xcompiler", "-fPIC,-O3", "--expt-relaxed-constexpr",
         "-Xptxas", "-warn-spills"] + os.environ.get("ACCEL_NVCC_EXTRA", "").split()


def sources() -> list[str]:
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")) + glob.glob(os.path.join(CSRC, "host", "*.cpp")))


def deps() -> list[str]:
    pats = ["*.cu", "*.cuh", "*.h", "*.cpp", "*/*.cu", "*/*.cuh", "*/*.h", "*/*.cpp"]
    out = [p for pat in pats for p in glob.glob(os.path.join(CSRC, pat))]
    return out + glob.glob(os.path.join(INCLUDE, "*.h")) + glob.glob(os.path.join(INCLUDE, "*.cuh")) + \
        glob.glob(os.path.join(ROOT, "examples", "*.cu"))


def up_to_date() -> bool:
    if not os.path.exists(LIB):
        return False
    t = os.path.getmtime(LIB)
    if not all(os.path.exists(p) for p in (LIB_RT, LIB_INTERCEPT)):
        return False
    return all(os.path.getmtime(p) <= t for p in deps())


def build(force: bool = False, verbose: bool = False) -> str:
    if not force and up_to_date():
        return LIB
    objdir = os.path.join(PKG, "build")
    os.makedirs(objdir, exist_ok=True)
    objs = []
    for src in sources():
        obj = os.path.join(objdir, os.path.basename(src) + ".o")
        cmd = [NVCC, *ARCH, *FLAGS, "-I", INCLUDE, "-I", CSRC, "-c", src, "-o", obj]
        if verbose and src.endswith(".cu"):
            cmd += ["-Xptxas", "-v"]
        subprocess.check_call(cmd)
        objs.append(obj)
    tmp = LIB + f".tmp{os.getpid()}"
    subprocess.check_call([NVCC, *ARCH, "-shared", "-cudart", "static", "-o", tmp, *objs,
                           "-Xcompiler", "-fPIC"])
    os.replace(tmp, LIB)
    build_intercept(objs)
    return LIB


def build_intercept(objs: list[str]) -> None:
    """Transparent interception: the same objects linked
    against the SHARED CUDA runtime (libaccel_rt.so: an application's kernel
    stubs and the library must live in one runtime instance), the LD_PRELOAD
    shim over cudaLaunchKernel (libaccel_intercept.so), and the example
    application (examples/intercept_app, shared runtime)."""
    tmp = LIB_RT + f".tmp{os.getpid()}"
    subprocess.check_call([NVCC, *ARCH, "-shared", "-cudart", "shared", "-o", tmp, *objs, "-Xcompiler", "-fPIC"])
    os.replace(tmp, LIB_RT)
    tmp = LIB_INTERCEPT + f".tmp{os.getpid()}"
    subprocess.check_call([NVCC, "-std=c++17", "-O2", "-shared", "-cudart", "shared", "-Xcompiler", "-fPIC",
                           "-I", INCLUDE, os.path.join(CSRC, "intercept", "intercept.cpp"), "-o", tmp,
                           "-L", PKG, "-laccel_rt", "-ldl", "-Xlinker", "-rpath,$ORIGIN"])
    os.replace(tmp, LIB_INTERCEPT)
    app_src = os.path.join(ROOT, "examples", "intercept_app.cu")
    if os.path.exists(app_src):
        tmp = APP + f".tmp{os.getpid()}"
        subprocess.check_call([NVCC, *ARCH, "-O2", "-std=c++17", "--expt-relaxed-constexpr", "-cudart", "shared",
                               "-I", INCLUDE, "-I", CSRC, app_src, "-o", tmp])
        os.replace(tmp, APP)


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose="--verbose" in sys.argv)
    print(LIB)

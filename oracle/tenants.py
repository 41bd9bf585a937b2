"""ctypes front end of liboracle (TEST INFRASTRUCTURE ONLY -- see oracle/__init__.py).

Each function takes the input dict produced by `synth` and returns the
tenant's reference outputs as numpy arrays.  No arithmetic happens here
beyond marshalling; the definitions live in oracle/tenants.c.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_HERE, "liboracle.so")
SRC_PATH = os.path.join(_HERE, "tenants.c")
CFLAGS = ["-O2", "-fopenmp", "-ffp-contract=off", "-fno-fast-math", "-fPIC", "-shared", "-std=c11"]


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (plain C, OpenMP, no FMA contraction)."""
    if force or not os.path.exists(LIB_PATH) or os.path.getmtime(LIB_PATH) < os.path.getmtime(SRC_PATH):
        tmp = LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", *CFLAGS, "-o", tmp, SRC_PATH, "-lm"])
        os.replace(tmp, LIB_PATH)
    return LIB_PATH


_lib = None


def lib() -> C.CDLL:
    global _lib
    if _lib is None:
        build()
        _lib = C.CDLL(LIB_PATH)
    return _lib


def _p(a: np.ndarray) -> C.c_void_p:
    assert a.flags["C_CONTIGUOUS"], "oracle needs contiguous arrays"
    return C.c_void_p(a.ctypes.data)


I64 = C.c_int64


def mop(d: dict) -> np.ndarray:
    out = np.empty(d["n"], dtype=np.float32)
    lib().oracle_mop(_p(d["ina"]), _p(d["inb"]), _p(out), I64(d["n"]), I64(d["block"]),
                     I64(d["nconst"]))
    return out


def stencil(d: dict) -> np.ndarray:
    out = np.empty((d["nz"], d["ny"], d["nx"]), dtype=np.float64)
    lib().oracle_stencil(_p(d["a0"]), _p(out), I64(d["nx"]), I64(d["ny"]), I64(d["nz"]),
                         I64(d["sweeps"]), C.c_double(d["c0"]), C.c_double(d["c1"]))
    return out


def histo(d: dict) -> tuple[np.ndarray, np.ndarray]:
    counts = np.empty(d["bins"], dtype=np.uint32)
    sat = np.empty(d["bins"], dtype=np.uint8)
    lib().oracle_histo(_p(d["samples"]), C.c_int(d["sample_bytes"]), I64(d["n"]), I64(d["bins"]),
                       _p(counts), _p(sat))
    return counts, sat


def bfs(d: dict) -> tuple[np.ndarray, int]:
    level = np.empty(d["nv"], dtype=np.int32)
    f = lib().oracle_bfs
    f.restype = C.c_int
    depth = f(_p(d["row_ptr"]), _p(d["col"]), I64(d["nv"]), I64(d["src"]), _p(level))
    return level, int(depth)


def cutcp(d: dict) -> np.ndarray:
    v = np.empty((d["nz"], d["ny"], d["nx"]), dtype=np.float64)
    lib().oracle_cutcp(_p(d["atoms"]), I64(d["natoms"]), I64(d["nx"]), I64(d["ny"]), I64(d["nz"]),
                       C.c_float(d["h"]), C.c_float(d["cutoff"]), C.c_float(d["excl"]), _p(v))
    return v


def cutcp_points(d: dict, ijk: np.ndarray) -> np.ndarray:
    ijk = np.ascontiguousarray(ijk, dtype=np.int32).reshape(-1, 3)
    v = np.empty(len(ijk), dtype=np.float64)
    lib().oracle_cutcp_points(_p(d["atoms"]), I64(d["natoms"]), _p(ijk), I64(len(ijk)),
                              C.c_float(d["h"]), C.c_float(d["cutoff"]), C.c_float(d["excl"]), _p(v))
    return v


def tpacf(d: dict) -> tuple[np.ndarray, np.ndarray, np.ndarray]:
    nb = len(d["binb"]) + 1
    dd = np.empty(nb, dtype=np.uint64)
    rr = np.empty(nb, dtype=np.uint64)
    dr = np.empty(nb, dtype=np.uint64)
    rc = lib().oracle_tpacf(_p(d["data"]), _p(d["rand"]), I64(d["npts"]), I64(d["nsets"]),
                            _p(d["binb"]), C.c_int(len(d["binb"])), _p(dd), _p(rr), _p(dr))
    assert rc == 0
    return dd, rr, dr


def spmv(d: dict) -> np.ndarray:
    y = np.empty(d["n"], dtype=np.float64)
    lib().oracle_spmv(_p(d["row_ptr"]), _p(d["col"]), _p(d["val"]), _p(d["x"]), I64(d["n"]), _p(y))
    return y


def sgemm(d: dict) -> np.ndarray:
    c = np.empty((d["m"], d["n"]), dtype=np.float64)
    lib().oracle_sgemm(_p(d["a"]), _p(d["b"]), I64(d["m"]), I64(d["n"]), I64(d["k"]), _p(c))
    return c


def sgemm_entries(d: dict, ij: np.ndarray) -> np.ndarray:
    ij = np.ascontiguousarray(ij, dtype=np.int64).reshape(-1, 2)
    c = np.empty(len(ij), dtype=np.float64)
    lib().oracle_sgemm_entries(_p(d["a"]), _p(d["b"]), I64(d["k"]), _p(ij), I64(len(ij)), _p(c))
    return c


def mriq_phimag(d: dict) -> np.ndarray:
    pm = np.empty(d["numk"], dtype=np.float32)
    lib().oracle_mriq_phimag(_p(d["phir"]), _p(d["phii"]), I64(d["numk"]), _p(pm))
    return pm


def mriq_points(d: dict, idx: np.ndarray, phimag: np.ndarray | None = None):
    if phimag is None:
        phimag = mriq_phimag(d)
    idx = np.ascontiguousarray(idx, dtype=np.int64)
    qr = np.empty(len(idx), dtype=np.float64)
    qi = np.empty(len(idx), dtype=np.float64)
    lib().oracle_mriq_points(_p(d["kx"]), _p(d["ky"]), _p(d["kz"]), _p(phimag), I64(d["numk"]),
                             _p(d["x"]), _p(d["y"]), _p(d["z"]), _p(idx), I64(len(idx)), _p(qr), _p(qi))
    return qr, qi


def mriq(d: dict):
    pm = mriq_phimag(d)
    qr, qi = mriq_points(d, np.arange(d["numx"]), pm)
    return pm, qr, qi


def sad(d: dict):
    """(sad4 u16[mb][p][16], sad8 u16[mb][p][4], sad16 u16[mb][p])."""
    nmb = (d["w"] // 16) * (d["h"] // 16)
    npos = (2 * d["R"] + 1) ** 2
    s4 = np.empty((nmb, npos, 16), dtype=np.uint16)
    s8 = np.empty((nmb, npos, 4), dtype=np.uint16)
    s16 = np.empty((nmb, npos), dtype=np.uint16)
    lib().oracle_sad(_p(d["cur"]), _p(d["ref"]), I64(d["w"]), I64(d["h"]), I64(d["R"]), _p(s4), _p(s8), _p(s16))
    return s4, s8, s16


def lbm(d: dict) -> np.ndarray:
    """f after `steps` stream-collide steps, float64 [19][nz][ny][nx]."""
    out = np.empty((19, d["nz"], d["ny"], d["nx"]), dtype=np.float64)
    lib().oracle_lbm(_p(d["f0"]), _p(d["flags"]), I64(d["nx"]), I64(d["ny"]), I64(d["nz"]), I64(d["steps"]),
                     C.c_double(d["omega"]), _p(out))
    return out


def histo_pipeline(d: dict):
    """(lo, hi, bin stream u32[n], counts u32[bins], sat u8[bins])."""
    n, bins = d["n"], d["bins"]
    lo, hi = C.c_uint32(), C.c_uint32()
    bo = np.empty(n, dtype=np.uint32)
    counts = np.empty(bins, dtype=np.uint32)
    sat = np.empty(bins, dtype=np.uint8)
    lib().oracle_histo_pipeline(_p(d["raw"]), I64(n), I64(bins), C.byref(lo), C.byref(hi), _p(bo), _p(counts), _p(sat))
    return lo.value, hi.value, bo, counts, sat


def gridding(d: dict) -> np.ndarray:
    """grid complex [G][G][G][2] float64 (re, im)."""
    G = d["G"]
    g = np.empty((G, G, G, 2), dtype=np.float64)
    lib().oracle_gridding(_p(d["x"]), _p(d["y"]), _p(d["z"]), _p(d["re"]), _p(d["im"]), I64(d["n"]), I64(G),
                          C.c_float(d["hw"]), _p(d["lut"]), I64(len(d["lut"])), _p(g))
    return g

"""Tenant jobs: device buffers + the accel_request a tenant submits.

Argument marshalling only.  Each Job uploads its seeded inputs (from `synth`)
into device memory owned by PyTorch, allocates outputs / scratch, and
describes its kernel execution request as steps of built-in kernels (names of
include/accel_tenants.h) -- the computation itself runs in libaccel.so.

A Job is one *request* in the sense of PAPER.md §7.2 (lines 853-860: "kernel
execution requests"); iterative Parboil codes submit their whole launch
sequence as one request (DESIGN.md R-job-1).
"""
from __future__ import annotations

import ctypes as C
import os
from dataclasses import dataclass, field

import numpy as np
import torch

from . import abi


def _dev(a: np.ndarray, device) -> torch.Tensor:
    a = np.ascontiguousarray(a)
    if a.dtype == np.uint32:
        a = a.view(np.int32)
    elif a.dtype == np.uint64:
        a = a.view(np.int64)
    return torch.from_numpy(a).to(device)


def _np(t: torch.Tensor, dtype) -> np.ndarray:
    return t.detach().cpu().numpy().view(dtype)


def _cdiv(a: int, b: int) -> int:
    return -(-a // b)


def _measured_peaks() -> dict:
    """MEASURED_PEAKS.json (driver-written, repo root); B200_PROFILING.md's
    fallback figures when it is absent."""
    import json
    import os
    p = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "MEASURED_PEAKS.json")
    try:
        with open(p) as f:
            return json.load(f)
    except OSError:
        return {"hbm_gbs": 6650.0, "bf16_tflops": 1590.0, "sm_max_mhz": 1965.0}


# Roofline peaks for the non-HBM tenants: FP32 SIMT derived from
# the guide's unit counts (148 SM x 128 FP32 lanes x 2 flop x max SM clock);
# TF32 tensor = the measured dense bf16 peak x the nominal TF32/BF16 ratio 1/2.
PEAKS = _measured_peaks()
FP32_SIMT_TFLOPS = 148 * 128 * 2 * PEAKS.get("sm_max_mhz", 1965.0) * 1e6 / 1e12
TF32_TENSOR_TFLOPS = PEAKS["bf16_tflops"] / 2


@dataclass
class Step:
    kernel: str
    grid: tuple[int, int, int]
    args: C.Structure
    repeat: int = 1
    order: torch.Tensor | None = None   # dequeue order (device uint32 permutation), None = linear


@dataclass
class Job:
    """Base class.  Subclasses fill `inputs` (device tensors the e2e path
    copies from host), `steps`, `clears` and `outputs`."""
    name: str = "job"
    device: torch.device = field(default_factory=lambda: torch.device("cuda"))

    def __post_init__(self):
        self.inputs: dict[str, torch.Tensor] = {}
        self.out: dict[str, torch.Tensor] = {}
        self.steps: list[Step] = []
        self.clears: list[tuple[torch.Tensor, int]] = []
        self._pinned_in: dict[str, torch.Tensor] = {}
        self._pinned_out: dict[str, torch.Tensor] = {}
        self.main_step = -1  # -1: the library picks the step with the most VGs

    # ---- e2e: host buffers ----------------------------------------------
    def pin_host(self) -> None:
        """Pinned host copies of the inputs (sources of the per-step H2D) and
        pinned output buffers (destinations of the D2H)."""
        for k, t in self.inputs.items():
            h = torch.empty(t.shape, dtype=t.dtype, pin_memory=True)
            h.copy_(t.cpu())
            self._pinned_in[k] = h
        for k, t in self.output_tensors().items():
            self._pinned_out[k] = torch.empty(t.shape, dtype=t.dtype, pin_memory=True)

    def h2d_bytes(self) -> int:
        return sum(t.numel() * t.element_size() for t in self.inputs.values())

    def d2h_bytes(self) -> int:
        return sum(t.numel() * t.element_size() for t in self.output_tensors().values())

    def output_tensors(self) -> dict[str, torch.Tensor]:
        return dict(self.out)

    # ---- the request ------------------------------------------------------
    def request(self, kernel_ids: dict[str, int], tenant: int, e2e: bool = False,
                weight: int = 1, flags: int = 0) -> abi.accel_request:
        steps = (abi.accel_launch * len(self.steps))()
        keep = []
        for i, s in enumerate(self.steps):
            steps[i] = abi.accel_launch(kernel_ids[s.kernel], abi.accel_dim3(*s.grid),
                                        C.cast(C.pointer(s.args), C.c_void_p), C.sizeof(s.args), s.repeat,
                                        s.order.data_ptr() if s.order is not None else None)
            keep.append(s.args)
        clears = (abi.accel_clear * max(1, len(self.clears)))()
        for i, (t, v) in enumerate(self.clears):
            clears[i] = abi.accel_clear(t.data_ptr(), v, t.numel() * t.element_size())
        h2d = (abi.accel_copy * max(1, len(self.inputs)))()
        d2h = (abi.accel_copy * max(1, len(self.out)))()
        nh = nd = 0
        if e2e:
            if not self._pinned_in:
                self.pin_host()
            for k, t in self.inputs.items():
                h = self._pinned_in[k]
                h2d[nh] = abi.accel_copy(t.data_ptr(), h.data_ptr(), t.numel() * t.element_size())
                nh += 1
            for k, t in self.output_tensors().items():
                h = self._pinned_out[k]
                d2h[nd] = abi.accel_copy(h.data_ptr(), t.data_ptr(), t.numel() * t.element_size())
                nd += 1
        req = abi.accel_request(tenant, flags, weight, self.main_step, len(self.steps), steps, len(self.clears), clears,
                                nh, h2d, nd, d2h)
        req._keep = (steps, clears, h2d, d2h, keep)  # keep ctypes buffers alive until submit
        return req

    def launches(self) -> int:
        return sum(s.repeat for s in self.steps)

    def kernels(self) -> list[str]:
        return sorted({s.kernel for s in self.steps})

    def result(self) -> dict[str, np.ndarray]:
        raise NotImplementedError

    def host_result(self) -> dict[str, np.ndarray]:
        """Outputs as read back by the e2e D2H copies."""
        raise NotImplementedError

    # algorithmic work of one request, for roofline figures
    def work(self) -> dict:
        return {}


class MopJob(Job):
    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="mop", device=torch.device(device))
        self.n, self.block = d["n"], d["block"]
        assert self.block == 256
        self.inputs = {"ina": _dev(d["ina"], self.device), "inb": _dev(d["inb"], self.device)}
        self.out = {"out": torch.empty(self.n, dtype=torch.float32, device=self.device)}
        self.args = abi.accel_mop_args(self.inputs["ina"].data_ptr(), self.inputs["inb"].data_ptr(),
                                       self.out["out"].data_ptr(), self.n, d["nconst"])
        self.steps = [Step("mop", (_cdiv(self.n, 256), 1, 1), self.args, 1)]

    def result(self):
        return {"out": _np(self.out["out"], np.float32)}

    def work(self):
        return {"bytes": 12 * self.n, "bound": "hbm"}


class StencilJob(Job):
    TX, TY, TZ = 128, 8, 8
    # nx % 4 == 0: cp.async staging ("stencil", the default) or TMA-staged
    # planes ("stencil_tma"); any nx: "stencil_x"
    KERNELS = ("stencil_tma", "stencil")

    def __init__(self, d: dict, device="cuda", kernel: str | None = None):
        super().__init__(name="stencil", device=torch.device(device))
        self.nx, self.ny, self.nz, self.sweeps = d["nx"], d["ny"], d["nz"], d["sweeps"]
        n = self.nx * self.ny * self.nz
        self.inputs = {"a0": _dev(d["a0"].ravel(), self.device)}
        self.buf = [torch.empty(n, dtype=torch.float32, device=self.device) for _ in range(2)]
        self.out = {"a": self.buf[(self.sweeps - 1) & 1]}
        self.args = abi.accel_stencil_args(self.inputs["a0"].data_ptr(), self.buf[0].data_ptr(),
                                           self.buf[1].data_ptr(), self.nx, self.ny, self.nz, d["c0"], d["c1"])
        # default: cp.async staging; stencil_tma is opt-in until its drift next to
        # bfs is understood (DESIGN.md §6 "stencil staging", scripts/diag_tma.py)
        kernel = kernel or d.get("kernel") or os.environ.get("ACCEL_STENCIL_KERNEL") or \
            ("stencil" if self.nx % 4 == 0 else "stencil_x")
        if kernel != "stencil_x" and self.nx % 4:
            raise ValueError(f"{kernel} needs nx % 4 == 0 (16-B rows); stencil_x takes any nx")
        if kernel in ("stencil_tma", "stencil_bulk"):
            # 3-D maps of a0, buf0, buf1: box = one staged plane (136 x 10 x 1)
            maps = b"".join(abi.accel_tma_map_3d(t.data_ptr(), self.nx, self.ny, self.nz, 136, 10, 1)
                            for t in (self.inputs["a0"], self.buf[0], self.buf[1]))
            self.args = abi.accel_stencil_tma_args((C.c_uint8 * 384).from_buffer_copy(maps), self.buf[0].data_ptr(),
                                                   self.buf[1].data_ptr(), self.nx, self.ny, self.nz,
                                                   d["c0"], d["c1"])
            self.args.a0 = self.inputs["a0"].data_ptr()
            self.args.l2hint = int(d.get("l2hint", os.environ.get("ACCEL_TMA_L2HINT", 0)))
            if d.get("tma_global_maps"):   # diagnostic (scripts/diag_tma.py)
                self.gmaps = torch.frombuffer(bytearray(maps), dtype=torch.uint8).to(self.device)
                self.args.gmaps = self.gmaps.data_ptr()
        self.kernel = kernel
        ty = 16 if kernel == "stencil2" else self.TY   # stencil2: two rows per warp
        tz = 16 if kernel == "stencil_z16" else self.TZ   # stencil_z16: 16 planes per VG
        grid = (_cdiv(self.nx, self.TX), _cdiv(self.ny, ty), _cdiv(self.nz, tz))
        self.steps = [Step(kernel, grid, self.args, self.sweeps)]

    def result(self):
        return {"a": _np(self.out["a"], np.float32).reshape(self.nz, self.ny, self.nx)}

    def work(self):
        pts = self.nx * self.ny * self.nz
        return {"bytes": 8 * pts * self.sweeps, "bytes_per_launch": 8 * pts, "bound": "hbm",
                "launches": self.sweeps}


class HistoJob(Job):
    def __init__(self, d: dict, device="cuda", samples: torch.Tensor | None = None):
        """samples: an existing device stream of bin indices (the histo
        pipeline's intermediates) instead of d["samples"]."""
        super().__init__(name="histo", device=torch.device(device))
        self.n, self.bins, self.iters, self.sb = d["n"], d["bins"], d["iters"], d["sample_bytes"]
        if not (1 <= self.bins <= 16384 and (self.sb == 4 or self.bins == 256)):
            raise ValueError("histo: 1..16384 bins; u8 samples need 256 bins")
        if self.n >= 1 << 32:
            raise ValueError("histo: n < 2^32 samples (u32 counters)")
        # > 4096 bins: the packed 16-bit private histogram (VGs < 65536 samples)
        self.kernel = "histo" if self.bins <= 4096 else "histo_wide"
        # samples per VG: histo_wide flushes up to 16K bins per VG with global
        # atomics, so its VGs are as large as the 16-bit counters allow
        # (measured at the SURVEY default: 74 -> 52 us per pass, 16384 -> 61440)
        self.per_vg = 4096 if self.sb == 1 else d.get("per_vg", 16384 if self.kernel == "histo" else 61440)
        assert self.per_vg % 4096 == 0 and (self.kernel == "histo" or self.per_vg < 65536)
        self.inputs = {"samples": _dev(d["samples"], self.device)} if samples is None else {}
        src = samples if samples is not None else self.inputs["samples"]
        self.hist = torch.zeros(2 * self.bins, dtype=torch.int32, device=self.device)
        self.sat = torch.zeros(self.bins, dtype=torch.uint8, device=self.device)
        self.done = torch.zeros(self.iters, dtype=torch.int32, device=self.device)
        last = (self.iters - 1) & 1
        self.out = {"counts": self.hist[last * self.bins:(last + 1) * self.bins], "sat": self.sat}
        self.args = abi.accel_histo_args(src.data_ptr(), self.n, self.bins, self.sb,
                                         self.per_vg, self.hist.data_ptr(), self.sat.data_ptr(),
                                         self.done.data_ptr())
        self.clears = [(self.hist, 0), (self.done, 0)]
        self.steps = [Step(self.kernel, (_cdiv(self.n, self.per_vg), 1, 1), self.args, self.iters)]

    def result(self):
        return {"counts": _np(self.out["counts"], np.uint32), "sat": _np(self.sat, np.uint8)}

    def work(self):
        b = self.n * self.sb + 4 * self.bins
        return {"bytes": b * self.iters, "bytes_per_launch": b, "bound": "hbm", "launches": self.iters}


class BfsJob(Job):
    """One request = `levels` launches of the level-expansion kernel (upper
    bound on the BFS depth; launches past the last level find an empty
    frontier on the device and return immediately)."""

    def __init__(self, d: dict, device="cuda", levels: int | None = None):
        super().__init__(name="bfs", device=torch.device(device))
        self.nv, self.ne, self.src = d["nv"], d["ne"], d["src"]
        self.levels = levels or d.get("levels", 24)
        self.inputs = {"row_ptr": _dev(d["row_ptr"], self.device), "col": _dev(d["col"], self.device)}
        self.level = torch.empty(self.nv, dtype=torch.int32, device=self.device)
        self.frontier = torch.empty(2 * self.nv, dtype=torch.int32, device=self.device)
        self.count = torch.zeros(self.levels + 1, dtype=torch.int32, device=self.device)
        self.out = {"level": self.level}
        self.args = abi.accel_bfs_args(self.inputs["row_ptr"].data_ptr(), self.inputs["col"].data_ptr(),
                                       self.nv, self.src, self.level.data_ptr(), self.frontier.data_ptr(),
                                       self.count.data_ptr())
        self.clears = [(self.level, 0xFF), (self.count, 0)]
        self.steps = [Step("bfs", (_cdiv(self.nv, 256), 1, 1), self.args, self.levels)]

    def result(self):
        return {"level": _np(self.level, np.int32)}

    def frontier_sizes(self):
        return _np(self.count, np.uint32)

    def set_levels(self, levels: int) -> None:
        """Re-size the request to `levels` level launches (same buffers)."""
        self.levels = int(levels)
        self.count = torch.zeros(self.levels + 1, dtype=torch.int32, device=self.device)
        self.args.count = self.count.data_ptr()
        self.clears = [(self.level, 0xFF), (self.count, 0)]
        self.steps = [Step("bfs", (_cdiv(self.nv, 256), 1, 1), self.args, self.levels)]

    def fit_levels(self, acc) -> int:
        """Parboil's bfs launches levels until the frontier is empty.  Here the
        whole launch sequence is one request (no host round trip per level),
        so its length is the graph's depth + 1, learned once by a probe run of
        this request through `acc` (untimed set-up, like knowing a stencil's
        sweep count): launch l writes the size of frontier l + 1 to count[l+1];
        the first empty one ends the search.  Returns the fitted launch count."""
        acc.run([self])
        c = self.frontier_sizes()
        empty = [l for l in range(1, len(c)) if c[l] == 0]
        if not empty:
            raise RuntimeError(f"bfs deeper than {self.levels} levels")
        self.set_levels(empty[0])
        return self.levels

    def work(self):
        b = 16 * self.nv + 8 * self.ne
        return {"bytes": b, "bytes_per_launch": b / self.levels, "bound": "hbm", "launches": self.levels}


class CutcpJob(Job):
    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="cutcp", device=torch.device(device))
        self.d = {k: d[k] for k in ("nx", "ny", "nz", "h", "cutoff", "excl", "natoms", "box")}
        self.nx, self.ny, self.nz = d["nx"], d["ny"], d["nz"]
        self.inputs = {"atoms": _dev(d["atoms"].ravel(), self.device),
                       "cell_start": _dev(d["cell_start"], self.device)}
        self.v = torch.empty(self.nz * self.ny * self.nx, dtype=torch.float32, device=self.device)
        self.out = {"v": self.v}
        self.args = abi.accel_cutcp_args(self.inputs["atoms"].data_ptr(), self.inputs["cell_start"].data_ptr(),
                                         d["ncell_1d"], d["cell"], self.nx, self.ny, self.nz, d["h"],
                                         d["cutoff"], d["excl"], self.v.data_ptr())
        grid = (_cdiv(self.nx, 8), _cdiv(self.ny, 8), _cdiv(self.nz, 8))
        # dequeue order: the library's cost model (Cutcp::vg_cost, most atoms first)
        self.steps = [Step("cutcp", grid, self.args, 1)]

    def result(self):
        return {"v": _np(self.v, np.float32).reshape(self.nz, self.ny, self.nx)}

    def work(self):
        # in-cutoff (lattice point, atom) pairs, estimated from the mean atom
        # density (cutcp algorithmic work); ~15 flop each
        dens = self.d["natoms"] / self.d["box"] ** 3
        pairs = self.nx * self.ny * self.nz * dens * 4.0 / 3.0 * np.pi * self.d["cutoff"] ** 3
        return {"pairs": pairs, "flops": 15.0 * pairs, "bound": "alu", "launches": 1, "peak_tflops": FP32_SIMT_TFLOPS}


class TpacfJob(Job):
    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="tpacf", device=torch.device(device))
        self.n, self.S = d["npts"], d["nsets"]
        self.nedges = len(d["binb"])
        assert self.nedges + 1 <= 32
        self.inputs = {"data": _dev(d["data"], self.device), "rand": _dev(d["rand"], self.device),
                       "binb": _dev(d["binb"], self.device)}
        nb = self.nedges + 1
        self.hists = torch.zeros(3 * nb, dtype=torch.int64, device=self.device)
        self.out = {"hists": self.hists}
        p = self.hists.data_ptr()
        # VGs split the other set's tiles in `qsplit` runs: finer VGs, shorter tail
        self.qsplit = int(d.get("qsplit", os.environ.get("ACCEL_TPACF_QSPLIT", 2)))
        self.args = abi.accel_tpacf_args(self.inputs["data"].data_ptr(), self.inputs["rand"].data_ptr(),
                                         self.inputs["binb"].data_ptr(), self.n, self.S, self.nedges, self.qsplit,
                                         p, p + 8 * nb, p + 16 * nb)
        self.clears = [(self.hists, 0)]
        grid = (_cdiv(self.n, 256), 2 * self.S + 1, self.qsplit)
        # dequeue order: the library's cost model (Tpacf::vg_cost, longest pair blocks first)
        self.steps = [Step("tpacf", grid, self.args, 1)]

    def result(self):
        h = _np(self.hists, np.uint64).reshape(3, -1)
        return {"dd": h[0], "rr": h[1], "dr": h[2]}

    def work(self):
        n, S = self.n, self.S
        pairs = (1 + S) * n * (n - 1) // 2 + S * n * n
        return {"pairs": pairs, "flops": 5.0 * pairs, "bound": "alu", "launches": 1, "peak_tflops": FP32_SIMT_TFLOPS}


class SpmvJob(Job):
    """kernel "spmv" (default) or "spmv_v4" (ACCEL_SPMV_KERNEL=spmv_v4: 128-bit
    chunk loads over col/val padded to a multiple of 4 elements).  spmv_v4 is
    22 % faster natively but only 7 % in SHARED mode (2-us VGs: the per-VG
    hand-over of the persistent loop shows), which made the sampled mixes less
    fair (its T(a) fell more than its shared time) -- DESIGN.md §6."""

    def __init__(self, d: dict, device="cuda", kernel: str | None = None):
        super().__init__(name="spmv", device=torch.device(device))
        self.n, self.nnz, self.iters = d["n"], d["nnz"], d["iters"]
        self.kernel = kernel or os.environ.get("ACCEL_SPMV_KERNEL", "spmv")
        pad = (-self.nnz) % 4 if self.kernel == "spmv_v4" else 0
        arrs = {k: d[k] for k in ("row_ptr", "col", "val", "x")}
        if pad:
            arrs["col"] = np.concatenate([arrs["col"], np.zeros(pad, arrs["col"].dtype)])
            arrs["val"] = np.concatenate([arrs["val"], np.zeros(pad, arrs["val"].dtype)])
        self.inputs = {k: _dev(v, self.device) for k, v in arrs.items()}
        self.y = torch.empty(self.n, dtype=torch.float32, device=self.device)
        self.out = {"y": self.y}
        i = self.inputs
        self.args = abi.accel_spmv_args(i["row_ptr"].data_ptr(), i["col"].data_ptr(), i["val"].data_ptr(),
                                        i["x"].data_ptr(), self.y.data_ptr(), self.n)
        self.steps = [Step(self.kernel, (_cdiv(self.n, 64), 1, 1), self.args, self.iters)]

    def result(self):
        return {"y": _np(self.y, np.float32)}

    def work(self):
        b = 8 * self.nnz + 12 * self.n
        return {"bytes": b * self.iters, "bytes_per_launch": b, "bound": "hbm", "launches": self.iters}


class SgemmJob(Job):
    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="sgemm", device=torch.device(device))
        self.m, self.n, self.k = d["m"], d["n"], d["k"]
        if self.k % 4:
            raise ValueError("sgemm needs k % 4 == 0 (16-B rows)")
        self.inputs = {"a": _dev(d["a"].ravel(), self.device), "b": _dev(d["b"].ravel(), self.device)}
        self.c = torch.empty(self.m * self.n, dtype=torch.float32, device=self.device)
        self.out = {"c": self.c}
        self.args = abi.accel_sgemm_args(self.inputs["a"].data_ptr(), self.inputs["b"].data_ptr(),
                                         self.c.data_ptr(), self.m, self.n, self.k)
        self.steps = [Step("sgemm", (_cdiv(self.n, 128), _cdiv(self.m, 128), 1), self.args, 1)]

    def result(self):
        return {"c": _np(self.c, np.float32).reshape(self.m, self.n)}

    def work(self):
        f = 2.0 * self.m * self.n * self.k
        return {"flops": f, "flops_per_launch": f, "bound": "alu", "launches": 1, "peak_tflops": FP32_SIMT_TFLOPS}


class SgemmTcJob(Job):
    """sgemm on the tcgen05 tensor cores (3xTF32).  k % 4 == 0 (16-B aligned
    rows for TMA): one step, sgemm_tc1, splitting hi/lo in shared memory;
    otherwise two steps, split(A and B) into padded hi/lo arrays, then tc.
    The one-step form is the default; one_step=False or
    ACCEL_SGEMM_ONESTEP=0 selects split + tc."""

    def __init__(self, d: dict, device="cuda", one_step=None):
        super().__init__(name="sgemm", device=torch.device(device))
        self.m, self.n, self.k = d["m"], d["n"], d["k"]
        self.inputs = {"a": _dev(d["a"].ravel(), self.device), "b": _dev(d["b"].ravel(), self.device)}
        m, n, k = self.m, self.n, self.k
        if one_step is None:
            one_step = os.environ.get("ACCEL_SGEMM_ONESTEP", "1") != "0"
        self.one_step = bool(one_step) and k % 4 == 0
        self.c = torch.empty(m * n, dtype=torch.float32, device=self.device)
        self.out = {"c": self.c}
        if self.one_step:
            maps = b"".join([
                abi.accel_tma_map_2d(self.inputs["a"].data_ptr(), k, m, 4 * k, 16, 128, swizzle=64),
                abi.accel_tma_map_2d(self.inputs["b"].data_ptr(), k, n, 4 * k, 16, 256, swizzle=64)])
            self.tmaps = torch.frombuffer(bytearray(maps), dtype=torch.uint8).to(self.device)
            self.args_tc = abi.accel_sgemm_tc_args(self.tmaps.data_ptr(), self.c.data_ptr(), m, n, k)
            self.main_step = 0
            self.steps = [Step("sgemm_tc1", (_cdiv(n, 256), _cdiv(m, 128), 1), self.args_tc, 1)]
            return
        kp = _cdiv(k, 4) * 4   # hi/lo row stride: 16-B aligned rows for TMA
        self.split = {x: torch.empty(sz, dtype=torch.float32, device=self.device)
                      for x, sz in (("a_hi", m * kp), ("a_lo", m * kp), ("b_hi", n * kp), ("b_lo", n * kp))}
        maps = b"".join([
            abi.accel_tma_map_2d(self.split["a_hi"].data_ptr(), k, m, 4 * kp, 32, 128),
            abi.accel_tma_map_2d(self.split["a_lo"].data_ptr(), k, m, 4 * kp, 32, 128),
            abi.accel_tma_map_2d(self.split["b_hi"].data_ptr(), k, n, 4 * kp, 32, 256),
            abi.accel_tma_map_2d(self.split["b_lo"].data_ptr(), k, n, 4 * kp, 32, 256)])
        self.tmaps = torch.frombuffer(bytearray(maps), dtype=torch.uint8).to(self.device)
        s = self.split
        # one launch splits both operands (VGs of A first, then of B)
        self.args_s = abi.accel_sgemm_split_args(self.inputs["a"].data_ptr(), s["a_hi"].data_ptr(),
                                                 s["a_lo"].data_ptr(), m * k,
                                                 self.inputs["b"].data_ptr(), s["b_hi"].data_ptr(),
                                                 s["b_lo"].data_ptr(), n * k, k, kp)
        self.args_tc = abi.accel_sgemm_tc_args(self.tmaps.data_ptr(), self.c.data_ptr(), m, n, k)
        self.main_step = 1
        self.steps = [Step("sgemm_split", (_cdiv(m * k, 4096) + _cdiv(n * k, 4096), 1, 1), self.args_s, 1),
                      Step("sgemm_tc", (_cdiv(n, 256), _cdiv(m, 128), 1), self.args_tc, 1)]

    def result(self):
        return {"c": _np(self.c, np.float32).reshape(self.m, self.n)}

    def work(self):
        f = 2.0 * self.m * self.n * self.k
        # roofline of the dominant (tc) launch: 3 tf32 products per algorithmic MAC
        return {"flops": f, "flops_per_launch": f, "bound": "tensor", "launches": len(self.steps),
                "skip_launches": len(self.steps) - 1, "mma_flops": 3 * f, "peak_tflops": TF32_TENSOR_TFLOPS}


class MriqJob(Job):
    """Two steps, like Parboil's mri-q: ComputePhiMag (tiny) then ComputeQ."""

    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="mriq", device=torch.device(device))
        self.numx, self.numk = d["numx"], d["numk"]
        self.inputs = {k: _dev(d[k], self.device) for k in ("kx", "ky", "kz", "phir", "phii", "x", "y", "z")}
        i = self.inputs
        self.phimag = torch.empty(self.numk, dtype=torch.float32, device=self.device)
        self.qr = torch.empty(self.numx, dtype=torch.float32, device=self.device)
        self.qi = torch.empty(self.numx, dtype=torch.float32, device=self.device)
        self.out = {"phimag": self.phimag, "qr": self.qr, "qi": self.qi}
        self.args_pm = abi.accel_mriq_phimag_args(i["phir"].data_ptr(), i["phii"].data_ptr(),
                                                  self.phimag.data_ptr(), self.numk)
        self.args_q = abi.accel_mriq_q_args(i["kx"].data_ptr(), i["ky"].data_ptr(), i["kz"].data_ptr(),
                                            self.phimag.data_ptr(), self.numk, self.numx, i["x"].data_ptr(),
                                            i["y"].data_ptr(), i["z"].data_ptr(), self.qr.data_ptr(),
                                            self.qi.data_ptr())
        self.main_step = 1
        self.steps = [Step("mriq_phimag", (_cdiv(self.numk, 256), 1, 1), self.args_pm, 1),
                      Step("mriq_q", (_cdiv(self.numx, 256), 1, 1), self.args_q, 1)]

    def result(self):
        return {k: _np(t, np.float32) for k, t in self.out.items()}

    def work(self):
        pairs = self.numx * self.numk
        return {"pairs": pairs, "flops": 11.0 * pairs, "sfu": 2 * pairs, "bound": "alu", "launches": 2,
                "skip_launches": 1, "flops_per_launch": 11.0 * pairs, "peak_tflops": FP32_SIMT_TFLOPS}


class SadJob(Job):
    """Parboil sad (f3): three steps -- 4x4 SADs over the search window, then
    the 8x8 and 16x16 sums -- one request (R-solver-8; main step = 4x4)."""

    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="sad", device=torch.device(device))
        self.w, self.h, self.R = d["w"], d["h"], d["R"]
        if self.w % 16 or self.h % 16 or not 0 <= self.R <= 16:
            raise ValueError("sad: w, h multiples of 16 and R <= 16")
        self.inputs = {"cur": _dev(d["cur"].view(np.int16), self.device),
                       "ref": _dev(d["ref"].view(np.int16), self.device)}
        nmb, npos = (self.w // 16) * (self.h // 16), (2 * self.R + 1) ** 2
        self.nmb, self.npos = nmb, npos
        self.s4 = torch.empty(nmb * npos * 16, dtype=torch.int16, device=self.device)
        self.s8 = torch.empty(nmb * npos * 4, dtype=torch.int16, device=self.device)
        self.s16 = torch.empty(nmb * npos, dtype=torch.int16, device=self.device)
        self.out = {"sad4": self.s4, "sad8": self.s8, "sad16": self.s16}
        self.args = abi.accel_sad_args(self.inputs["cur"].data_ptr(), self.inputs["ref"].data_ptr(),
                                       self.s4.data_ptr(), self.s8.data_ptr(), self.s16.data_ptr(),
                                       self.w, self.h, self.R)
        grid = (self.w // 16, self.h // 16, 1)
        self.main_step = 0
        self.steps = [Step("sad_4x4", grid, self.args, 1), Step("sad_8x8", grid, self.args, 1),
                      Step("sad_16x16", grid, self.args, 1)]

    def result(self):
        return {"sad4": _np(self.s4, np.uint16).reshape(self.nmb, self.npos, 16),
                "sad8": _np(self.s8, np.uint16).reshape(self.nmb, self.npos, 4),
                "sad16": _np(self.s16, np.uint16).reshape(self.nmb, self.npos)}

    def work(self):
        # the dominant (4x4) launch: 256 absolute differences per (macroblock, displacement)
        n = self.nmb * self.npos
        return {"ops": 256 * n, "bytes": 2 * 16 * n + 4 * self.w * self.h, "bound": "alu", "launches": 3,
                "skip_launches": 0, "flops_per_launch": 2.0 * 256 * n, "peak_tflops": FP32_SIMT_TFLOPS}


class HistoPipelineJob(Job):
    """Parboil histo's whole pipeline (f3): prescan (input range), intermediates
    (raw samples -> bin indices), then `iters` launches of the main+final
    kernel on the bin stream -- one request, three steps (main = the last)."""

    # samples per VG of the prescan and intermediates steps: 4096 gives 4096
    # VGs for 2^24 samples, several waves over the persistent grid (16384
    # left 1024 VGs for 888 CTAs: a second wave of 136 -- +3.9 % STATIC; sweep
    # in profiles/r2b/histo_pipeline_per_vg.log)
    PER_VG = 4096

    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="histo_pipeline", device=torch.device(device))
        self.n, self.bins, self.iters = d["n"], d["bins"], d["iters"]
        self.PER_VG = int(d.get("per_vg", os.environ.get("ACCEL_HISTO_PRE_PER_VG", self.PER_VG)))
        self.inputs = {"raw": _dev(d["raw"], self.device)}
        self.bin_stream = torch.empty(self.n, dtype=torch.int32, device=self.device)
        self.lo = torch.empty(1, dtype=torch.int32, device=self.device)
        self.hi = torch.empty(1, dtype=torch.int32, device=self.device)
        self.main = HistoJob({"n": self.n, "bins": self.bins, "iters": self.iters, "sample_bytes": 4,
                              "samples": np.zeros(0, dtype=np.uint32)}, device, samples=self.bin_stream)
        self.hist, self.sat = self.main.hist, self.main.sat
        self.out = dict(self.main.out, lo=self.lo, hi=self.hi)
        self.args_pre = abi.accel_histo_pre_args(self.inputs["raw"].data_ptr(), self.bin_stream.data_ptr(),
                                                 self.lo.data_ptr(), self.hi.data_ptr(), self.n, self.bins,
                                                 self.PER_VG)
        self.clears = [(self.lo, 0xFF), (self.hi, 0)] + self.main.clears
        g = (_cdiv(self.n, self.PER_VG), 1, 1)
        self.main_step = 2
        self.steps = [Step("histo_prescan", g, self.args_pre, 1), Step("histo_intermediates", g, self.args_pre, 1),
                      self.main.steps[0]]

    def result(self):
        r = self.main.result()
        r.update(lo=int(_np(self.lo, np.uint32)[0]), hi=int(_np(self.hi, np.uint32)[0]))
        return r

    def work(self):
        b = 4 * self.n
        return {"bytes": 3 * b + self.main.work()["bytes"], "bound": "hbm", "launches": 2 + self.iters}


class GriddingJob(Job):
    """Parboil mri-gridding (f3): six steps -- binning, the three-kernel scan
    of the cell counts, reorder, gridding -- one request (main = gridding)."""

    CELL = 2.0   # cell edge in grid units: the gridding VG reads the cells within hw of its 8^3 tile

    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="gridding", device=torch.device(device))
        self.n, self.G, self.hw = d["n"], d["G"], d["hw"]
        dev = self.device
        self.inputs = {k: _dev(d[k], dev) for k in ("x", "y", "z", "re", "im", "lut")}
        self.cells = _cdiv(self.G, int(self.CELL))
        B = self.cells ** 3
        if B > 1024 * 1024 or len(d["lut"]) > 1024:
            raise ValueError("gridding: at most 1024^2 cells and 1024 LUT entries")
        u32 = lambda m: torch.empty(m, dtype=torch.int32, device=dev)  # noqa: E731
        f32 = lambda m: torch.empty(m, dtype=torch.float32, device=dev)  # noqa: E731
        self.bin, self.rank, self.count, self.start = u32(self.n), u32(self.n), u32(B), u32(B + 1)
        self.block_sum = u32(_cdiv(B, 1024))
        self.sorted = [f32(self.n) for _ in range(5)]
        self.grid = f32(2 * self.G ** 3)
        self.out = {"grid": self.grid}
        i = self.inputs
        self.args = abi.accel_gridding_args(i["x"].data_ptr(), i["y"].data_ptr(), i["z"].data_ptr(),
                                            i["re"].data_ptr(), i["im"].data_ptr(), i["lut"].data_ptr(),
                                            len(d["lut"]), self.n, self.G, self.cells, self.hw, self.CELL,
                                            self.bin.data_ptr(), self.rank.data_ptr(), self.count.data_ptr(),
                                            self.start.data_ptr(), self.block_sum.data_ptr(),
                                            *[t.data_ptr() for t in self.sorted], self.grid.data_ptr())
        self.clears = [(self.count, 0)]
        gs, gb = (_cdiv(self.n, 1024), 1, 1), (_cdiv(B, 1024), 1, 1)
        t = _cdiv(self.G, 8)
        self.main_step = 5
        self.steps = [Step("gridding_binning", gs, self.args), Step("gridding_scan_l1", gb, self.args),
                      Step("gridding_scan_inter", (1, 1, 1), self.args), Step("gridding_scan_add", gb, self.args),
                      Step("gridding_reorder", gs, self.args), Step("gridding_grid", (t, t, t), self.args)]

    def result(self):
        return {"grid": _np(self.grid, np.float32).reshape(self.G, self.G, self.G, 2)}

    def work(self):
        return {"bytes": 4 * 8 * self.G ** 3 + 20 * self.n, "bound": "alu", "launches": 6}


class LbmJob(Job):
    """Parboil lbm (f3): `steps` launches of the D3Q19 stream-collide step,
    ping-pong buffers (like stencil); the result is buf[(steps-1)&1]."""

    def __init__(self, d: dict, device="cuda"):
        super().__init__(name="lbm", device=torch.device(device))
        self.nx, self.ny, self.nz, self.nsteps = d["nx"], d["ny"], d["nz"], d["steps"]
        n = self.nx * self.ny * self.nz
        self.inputs = {"f0": _dev(d["f0"].ravel(), self.device), "flags": _dev(d["flags"].ravel().view(np.int8), self.device)}
        self.buf = [torch.empty(19 * n, dtype=torch.float32, device=self.device) for _ in range(2)]
        self.out = {"f": self.buf[(self.nsteps - 1) & 1]}
        self.args = abi.accel_lbm_args(self.inputs["f0"].data_ptr(), self.buf[0].data_ptr(), self.buf[1].data_ptr(),
                                       self.inputs["flags"].data_ptr(), self.nx, self.ny, self.nz, d["omega"])
        self.steps = [Step("lbm", (_cdiv(self.nx, 128), self.ny, self.nz), self.args, self.nsteps)]

    def result(self):
        return {"f": _np(self.out["f"], np.float32).reshape(19, self.nz, self.ny, self.nx)}

    def work(self):
        b = (19 * 8 + 1) * self.nx * self.ny * self.nz
        return {"bytes": b * self.nsteps, "bytes_per_launch": b, "bound": "hbm", "launches": self.nsteps}


JOBS = {"mop": MopJob, "stencil": StencilJob, "histo": HistoJob, "bfs": BfsJob, "cutcp": CutcpJob,
        "tpacf": TpacfJob, "spmv": SpmvJob, "sgemm": SgemmTcJob, "sgemm_simt": SgemmJob, "mriq": MriqJob, "sad": SadJob, "lbm": LbmJob,
        "histo_pipeline": HistoPipelineJob, "gridding": GriddingJob}


def make_job(name: str, d: dict, device="cuda") -> Job:
    return JOBS[name](d, device)

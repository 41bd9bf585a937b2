"""ctypes binding of libaccel.so (include/accel.h, include/accel_tenants.h).

Argument marshalling only: every function here forwards to the C ABI with the
same name.  There is no Python or CPU fallback -- if the library is missing the
import fails loudly (build it with `python -m paper_conf_cgo_margiolaso16_b200.build`).
"""
from __future__ import annotations

import ctypes as C
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
# ACCEL_LIB: load another build of the same ABI (A/B measurements only)
LIB_PATH = os.environ.get("ACCEL_LIB") or os.path.join(_HERE, "libaccel.so")

ACCEL_OK = 0
ACCEL_EINVAL = -1
ACCEL_ENOFIT = -2
ACCEL_ECUDA = -3
ACCEL_ESTATE = -4
ACCEL_ECOVERAGE = -5
ACCEL_ENOMEM = -6
ACCEL_ENOTREADY = -7
ERRORS = {0: "ACCEL_OK", -1: "ACCEL_EINVAL", -2: "ACCEL_ENOFIT", -3: "ACCEL_ECUDA",
          -4: "ACCEL_ESTATE", -5: "ACCEL_ECOVERAGE", -6: "ACCEL_ENOMEM", -7: "ACCEL_ENOTREADY"}
MODE_NATIVE, MODE_SHARED = 0, 1
POLICY_STATIC, POLICY_RESOLVE = 0, 1
ACCEL_ALL = 2**64 - 1
MAX_TENANTS = 16
MAX_STEPS = 8
REQ_LAUNCH_EVENTS = 1
REQ_TRACE = 2
REQ_LINEAR_ORDER = 4

u32, i32, u64, f32, f64, vp = C.c_uint32, C.c_int32, C.c_uint64, C.c_float, C.c_double, C.c_void_p


class accel_dim3(C.Structure):
    _fields_ = [("x", u32), ("y", u32), ("z", u32)]


class accel_caps(C.Structure):
    _fields_ = [("sms", i32), ("thr_per_sm", i32), ("regs_per_sm", i32), ("smem_per_sm", i32),
                ("ctas_per_sm", i32)]


class accel_config(C.Structure):
    _fields_ = [("device", i32), ("mode", i32), ("policy", i32), ("verify", i32), ("caps", accel_caps)]


class accel_kernel_desc(C.Structure):
    _fields_ = [("name", C.c_char_p), ("persistent_fn", vp), ("persistent_resolve_fn", vp), ("native_fn", vp),
                ("topup_fn", vp),
                ("block", accel_dim3),
                ("dyn_smem", u32), ("regs", i32), ("chunk", u32), ("args_size", u32), ("order_fn", vp),
                ("max_ctas_per_sm", u32), ("slices", u32)]


class accel_kernel_info(C.Structure):
    _fields_ = [("thr", u32), ("regs", u32), ("smem", u32), ("cta", u32), ("num_regs", i32),
                ("static_smem", i32), ("occ_persistent", i32), ("occ_native", i32)]


class accel_launch(C.Structure):
    _fields_ = [("kernel_id", i32), ("grid", accel_dim3), ("args", vp), ("args_size", u32), ("repeat", u32),
                ("order_device", vp)]


class accel_clear(C.Structure):
    _fields_ = [("dst_device", vp), ("value", i32), ("bytes", u64)]


class accel_copy(C.Structure):
    _fields_ = [("dst", vp), ("src", vp), ("bytes", u64)]


class accel_request(C.Structure):
    _fields_ = [("tenant", i32), ("flags", u32), ("weight", u32), ("main_step", i32), ("n_steps", u32), ("steps", C.POINTER(accel_launch)),
                ("n_clear", u32), ("clear", C.POINTER(accel_clear)), ("n_h2d", u32),
                ("h2d", C.POINTER(accel_copy)), ("n_d2h", u32), ("d2h", C.POINTER(accel_copy))]


class accel_req_stats(C.Structure):
    _fields_ = [("first_start_ns", u64), ("last_end_ns", u64), ("elapsed_ms", f32), ("arrival_ms", f32),
                ("done_ms", f32), ("vgs_total", u32), ("launches", u32), ("quota_initial", u32),
                ("quota_min", u32), ("quota_max", u32), ("resolves", u32), ("max_ctas", u32),
                ("coverage_ok", i32), ("mode", i32)]


class accel_launch_stat(C.Structure):
    _fields_ = [("t_first_ns", u64), ("t_last_ns", u64), ("ctas_started", u32), ("max_alive", u32),
                ("total", u32), ("topped", u32)]


class accel_vg_record(C.Structure):
    _fields_ = [("t_start_ns", u64), ("t_end_ns", u64), ("sm", u32), ("cta", u32)]


class accel_demand(C.Structure):
    _fields_ = [("thr", u32), ("regs", u32), ("smem", u32), ("cta", u32), ("grid_vgs", u32), ("weight", u32)]


class accel_mix_metrics(C.Structure):
    _fields_ = [("unfairness", f64), ("stp", f64), ("antt", f64), ("is_max", f64), ("is_min", f64)]


# ---- tenant argument structs (include/accel_tenants.h) ---------------------
class accel_mop_args(C.Structure):
    _fields_ = [("ina", vp), ("inb", vp), ("out", vp), ("n", u32), ("nconst", u32)]


class accel_stencil_args(C.Structure):
    _fields_ = [("a0", vp), ("buf0", vp), ("buf1", vp), ("nx", u32), ("ny", u32), ("nz", u32),
                ("c0", f32), ("c1", f32)]


class accel_stencil_tma_args(C.Structure):
    # three 128-B CUtensorMaps first; the C struct is 64-B aligned, so its
    # size is rounded up to a multiple of 64 (trailing pad)
    _fields_ = [("tmaps", C.c_uint8 * 384), ("buf0", vp), ("buf1", vp), ("nx", u32), ("ny", u32), ("nz", u32),
                ("c0", f32), ("c1", f32), ("l2hint", u32), ("gmaps", vp), ("a0", vp), ("dbg", vp)]


class accel_histo_args(C.Structure):
    _fields_ = [("samples", vp), ("n", u32), ("bins", u32), ("sample_bytes", u32), ("per_vg", u32),
                ("hist", vp), ("sat", vp), ("done", vp)]


class accel_bfs_args(C.Structure):
    _fields_ = [("row_ptr", vp), ("col", vp), ("nv", u32), ("src", u32), ("level", vp),
                ("frontier", vp), ("count", vp)]


class accel_cutcp_args(C.Structure):
    _fields_ = [("atoms", vp), ("cell_start", vp), ("ncell", u32), ("cell", f32), ("nx", u32),
                ("ny", u32), ("nz", u32), ("h", f32), ("cutoff", f32), ("excl", f32), ("v", vp)]


class accel_tpacf_args(C.Structure):
    _fields_ = [("data", vp), ("rand", vp), ("binb", vp), ("npts", u32), ("nsets", u32),
                ("nedges", u32), ("qsplit", u32), ("dd", vp), ("rr", vp), ("dr", vp)]


class accel_spmv_args(C.Structure):
    _fields_ = [("row_ptr", vp), ("col", vp), ("val", vp), ("x", vp), ("y", vp), ("n", u32)]


class accel_sgemm_args(C.Structure):
    _fields_ = [("a", vp), ("b", vp), ("c", vp), ("m", u32), ("n", u32), ("k", u32)]


class accel_sgemm_split_args(C.Structure):
    _fields_ = [("src0", vp), ("hi0", vp), ("lo0", vp), ("n0", u64),
                ("src1", vp), ("hi1", vp), ("lo1", vp), ("n1", u64), ("cols", u32), ("ld", u32)]


class accel_sgemm_tc_args(C.Structure):
    _fields_ = [("tmaps", vp), ("c", vp), ("m", u32), ("n", u32), ("k", u32)]


# kernel variants that take the same argument struct
accel_stencil_x_args = accel_stencil_args
accel_sgemm_tc1_args = accel_sgemm_tc_args
accel_spmv_v4_args = accel_spmv_args
accel_stencil_deep_args = accel_stencil_args
accel_stencil2_args = accel_stencil_args
accel_stencil_z16_args = accel_stencil_args
accel_stencil_bulk_args = accel_stencil_tma_args
accel_histo_wide_args = accel_histo_args


class accel_histo_pre_args(C.Structure):
    _fields_ = [("raw", vp), ("bins_out", vp), ("lo", vp), ("hi", vp), ("n", u32), ("bins", u32), ("per_vg", u32)]


accel_histo_prescan_args = accel_histo_intermediates_args = accel_histo_pre_args


class accel_gridding_args(C.Structure):
    _fields_ = [("x", vp), ("y", vp), ("z", vp), ("re", vp), ("im", vp), ("lut", vp),
                ("L", u32), ("n", u32), ("G", u32), ("cells", u32), ("hw", f32), ("cell", f32),
                ("bin", vp), ("rank", vp), ("count", vp), ("start", vp), ("block_sum", vp),
                ("sx", vp), ("sy", vp), ("sz", vp), ("sre", vp), ("sim", vp), ("grid", vp)]


accel_gridding_binning_args = accel_gridding_scan_l1_args = accel_gridding_scan_inter_args = accel_gridding_args
accel_gridding_scan_add_args = accel_gridding_reorder_args = accel_gridding_grid_args = accel_gridding_args


class accel_lbm_args(C.Structure):
    _fields_ = [("f0", vp), ("buf0", vp), ("buf1", vp), ("flags", vp), ("nx", u32), ("ny", u32), ("nz", u32),
                ("omega", f32)]


class accel_sad_args(C.Structure):
    _fields_ = [("cur", vp), ("ref", vp), ("sad4", vp), ("sad8", vp), ("sad16", vp), ("w", u32), ("h", u32), ("R", u32)]


accel_sad_4x4_args = accel_sad_8x8_args = accel_sad_16x16_args = accel_sad_args


class accel_mriq_phimag_args(C.Structure):
    _fields_ = [("phir", vp), ("phii", vp), ("phimag", vp), ("numk", u32)]


class accel_mriq_q_args(C.Structure):
    _fields_ = [("kx", vp), ("ky", vp), ("kz", vp), ("phimag", vp), ("numk", u32), ("numx", u32),
                ("x", vp), ("y", vp), ("z", vp), ("qr", vp), ("qi", vp)]


EXPORTS = [
    "accel_init", "accel_finalize", "accel_set_mode", "accel_last_error", "accel_builtin_kernel",
    "accel_builtin_count", "accel_builtin_name", "accel_kernel_register", "accel_kernel_info_get",
    "accel_submit", "accel_submit_group", "accel_sync", "accel_epoch", "accel_stats", "accel_release",
    "accel_tenant_stream", "accel_launch_times", "accel_launch_stats", "accel_vg_trace", "accel_demand_of", "accel_solve", "accel_placement_order", "accel_dequeue_order", "accel_metrics", "accel_metrics_weighted", "accel_guided_weights", "accel_overlap", "accel_tma_map_2d", "accel_tma_map_3d",
]


class AccelError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"{ERRORS.get(code, code)}: {msg}")
        self.code = code


def _load() -> C.CDLL:
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"{LIB_PATH} is missing: build it with "
                          "`python -m paper_conf_cgo_margiolaso16_b200.build` (no CPU fallback exists)")
    lib = C.CDLL(LIB_PATH)
    P = C.POINTER
    sig = {
        "accel_init": (i32, [P(accel_config), P(vp)]),
        "accel_finalize": (i32, [vp]),
        "accel_set_mode": (i32, [vp, i32, i32]),
        "accel_last_error": (C.c_char_p, [vp]),
        "accel_builtin_kernel": (i32, [C.c_char_p, P(accel_kernel_desc)]),
        "accel_builtin_count": (i32, []),
        "accel_builtin_name": (C.c_char_p, [i32]),
        "accel_kernel_register": (i32, [vp, P(accel_kernel_desc), P(i32)]),
        "accel_kernel_info_get": (i32, [vp, i32, P(accel_kernel_info)]),
        "accel_submit": (i32, [vp, P(accel_request), P(u64)]),
        "accel_submit_group": (i32, [vp, u32, P(accel_request), P(u64)]),
        "accel_sync": (i32, [vp, u64]),
        "accel_epoch": (i32, [vp]),
        "accel_stats": (i32, [vp, u64, P(accel_req_stats)]),
        "accel_release": (i32, [vp, u64]),
        "accel_tenant_stream": (i32, [vp, i32, P(vp), P(vp)]),
        "accel_launch_times": (i32, [vp, u64, P(f32), u32, P(u32)]),
        "accel_launch_stats": (i32, [vp, u64, P(accel_launch_stat), u32, P(u32)]),
        "accel_vg_trace": (i32, [vp, u64, P(accel_vg_record), u64, P(u64)]),
        "accel_demand_of": (i32, [P(accel_caps), u32, u32, u32, u32, u32, P(accel_demand)]),
        "accel_solve": (i32, [P(accel_caps), P(accel_demand), i32, P(u32)]),
        "accel_placement_order": (i32, [P(accel_caps), P(accel_demand), i32, P(i32)]),
        "accel_dequeue_order": (i32, [vp, i32, P(accel_dim3), vp, u32, vp]),
        "accel_metrics_weighted": (i32, [P(f64), P(f64), P(f64), i32, P(f64), P(f64)]),
        "accel_guided_weights": (i32, [i32, i32, P(f64), P(f64), u32, P(u32), P(f64)]),
        "accel_metrics": (i32, [P(f64), P(f64), i32, P(accel_mix_metrics)]),
        "accel_overlap": (i32, [P(f64), P(f64), i32, P(f64)]),
        "accel_tma_map_2d": (i32, [vp, vp, u64, u64, u64, u32, u32, i32]),
        "accel_tma_map_3d": (i32, [vp, vp, u64, u64, u64, u32, u32, u32]),
    }
    for name, (res, args) in sig.items():
        fn = getattr(lib, name)
        fn.restype = res
        fn.argtypes = args
    return lib


lib = _load()


def check(rc: int, ctx=None) -> int:
    if rc != ACCEL_OK:
        msg = lib.accel_last_error(ctx)
        raise AccelError(rc, msg.decode() if msg else "")
    return rc


# ---- thin wrappers with the C names ---------------------------------------
def accel_init(device: int = 0, mode: int = MODE_SHARED, policy: int = POLICY_STATIC, verify: bool = False,
               caps: accel_caps | None = None) -> C.c_void_p:
    cfg = accel_config(device, mode, policy, int(verify), caps or accel_caps())
    ctx = vp()
    check(lib.accel_init(C.byref(cfg), C.byref(ctx)), None)
    return ctx


def accel_finalize(ctx) -> None:
    check(lib.accel_finalize(ctx))


def accel_set_mode(ctx, mode: int, policy: int = POLICY_STATIC) -> None:
    check(lib.accel_set_mode(ctx, mode, policy), ctx)


def accel_builtin_kernel(name: str) -> accel_kernel_desc:
    d = accel_kernel_desc()
    check(lib.accel_builtin_kernel(name.encode(), C.byref(d)))
    return d


def accel_builtin_names() -> list[str]:
    return [lib.accel_builtin_name(i).decode() for i in range(lib.accel_builtin_count())]


def accel_kernel_register(ctx, desc: accel_kernel_desc) -> int:
    kid = i32()
    check(lib.accel_kernel_register(ctx, C.byref(desc), C.byref(kid)), ctx)
    return kid.value


def accel_kernel_info_get(ctx, kid: int) -> accel_kernel_info:
    info = accel_kernel_info()
    check(lib.accel_kernel_info_get(ctx, kid, C.byref(info)), ctx)
    return info


def accel_submit_group(ctx, reqs: list[accel_request]) -> list[int]:
    arr = (accel_request * len(reqs))(*reqs)
    ids = (u64 * len(reqs))()
    check(lib.accel_submit_group(ctx, len(reqs), arr, ids), ctx)
    return list(ids)


def accel_submit(ctx, req: accel_request) -> int:
    return accel_submit_group(ctx, [req])[0]


def accel_sync(ctx, request_id: int = ACCEL_ALL) -> None:
    check(lib.accel_sync(ctx, request_id), ctx)


def accel_epoch(ctx) -> None:
    check(lib.accel_epoch(ctx), ctx)


def accel_stats(ctx, request_id: int) -> accel_req_stats:
    s = accel_req_stats()
    check(lib.accel_stats(ctx, request_id, C.byref(s)), ctx)
    return s


def accel_launch_times(ctx, request_id: int, n: int) -> list[float]:
    buf = (f32 * max(n, 1))()
    got = u32()
    check(lib.accel_launch_times(ctx, request_id, buf, n, C.byref(got)), ctx)
    return list(buf)[:got.value]


def accel_launch_stats(ctx, request_id: int, n: int) -> list[accel_launch_stat]:
    buf = (accel_launch_stat * max(n, 1))()
    got = u32()
    check(lib.accel_launch_stats(ctx, request_id, buf, n, C.byref(got)), ctx)
    return list(buf)[:got.value]


def accel_vg_trace(ctx, request_id: int):
    """All VG records of a request submitted with REQ_TRACE, as a numpy
    structured array (t_start_ns, t_end_ns, sm, cta)."""
    import numpy as np
    got = u64()
    check(lib.accel_vg_trace(ctx, request_id, None, 0, C.byref(got)), ctx)
    arr = np.zeros(got.value, dtype=[("t_start_ns", "<u8"), ("t_end_ns", "<u8"), ("sm", "<u4"), ("cta", "<u4")])
    if got.value:
        check(lib.accel_vg_trace(ctx, request_id, arr.ctypes.data_as(C.POINTER(accel_vg_record)), got.value, C.byref(got)), ctx)
    return arr


def accel_dequeue_order(ctx, kernel_id: int, grid, args: C.Structure, order_device_ptr: int) -> None:
    """The library's cost-model dequeue order for (kernel, grid, args) into a
    device uint32 buffer of G entries (synchronous)."""
    check(lib.accel_dequeue_order(ctx, kernel_id, C.byref(accel_dim3(*grid)), C.cast(C.pointer(args), C.c_void_p),
                                  C.sizeof(args), C.c_void_p(order_device_ptr)), ctx)


def accel_release(ctx, request_id: int = ACCEL_ALL) -> None:
    check(lib.accel_release(ctx, request_id), ctx)


def accel_tenant_stream(ctx, tenant: int) -> tuple[int, int]:
    a, b = vp(), vp()
    check(lib.accel_tenant_stream(ctx, tenant, C.byref(a), C.byref(b)), ctx)
    return a.value or 0, b.value or 0


def accel_demand_of(block: int, regs: int, smem: int, grid_vgs: int, weight: int = 1,
                    caps: accel_caps | None = None) -> accel_demand:
    d = accel_demand()
    check(lib.accel_demand_of(C.byref(caps or accel_caps()), block, regs, smem, grid_vgs, weight, C.byref(d)))
    return d


def accel_solve(demands: list[accel_demand], caps: accel_caps | None = None) -> list[int]:
    k = len(demands)
    arr = (accel_demand * max(k, 1))(*demands)
    out = (u32 * max(k, 1))()
    check(lib.accel_solve(C.byref(caps or accel_caps()), arr, k, out))
    return list(out)[:k]


def accel_placement_order(demands: list[accel_demand], caps: accel_caps | None = None) -> list[int]:
    """R-place-1: request indices, largest per-CTA footprint first."""
    k = len(demands)
    arr = (accel_demand * max(k, 1))(*demands)
    out = (i32 * max(k, 1))()
    check(lib.accel_placement_order(C.byref(caps or accel_caps()), arr, k, out))
    return list(out)[:k]



def accel_metrics(ta: list[float], ts: list[float]) -> accel_mix_metrics:
    k = len(ta)
    m = accel_mix_metrics()
    check(lib.accel_metrics((f64 * k)(*ta), (f64 * k)(*ts), k, C.byref(m)))
    return m


def accel_tma_map_2d(gaddr: int, inner: int, outer: int, row_stride_bytes: int, box_inner: int,
                     box_outer: int, swizzle: int = 128) -> bytes:
    out = (C.c_ubyte * 128)()
    check(lib.accel_tma_map_2d(out, gaddr, inner, outer, row_stride_bytes, box_inner, box_outer, swizzle))
    return bytes(out)


def accel_tma_map_3d(gaddr: int, d0: int, d1: int, d2: int, box0: int, box1: int, box2: int) -> bytes:
    out = (C.c_ubyte * 128)()
    check(lib.accel_tma_map_3d(out, gaddr, d0, d1, d2, box0, box1, box2))
    return bytes(out)


def accel_metrics_weighted(ta: list[float], ts: list[float], w: list[float]) -> tuple[float, list[float]]:
    """(weighted unfairness, weighted slowdowns) of one mix (DESIGN.md R-metric-5)."""
    k = len(ta)
    arr = lambda xs: (f64 * max(k, 1))(*xs)  # noqa: E731
    wu = f64()
    ws = (f64 * max(k, 1))()
    check(lib.accel_metrics_weighted(arr(ta), arr(ts), arr(w), k, C.byref(wu), ws))
    return wu.value, list(ws)[:k]


def accel_guided_weights(fracs: list[float], ms: list[list[float]], scale: int = 16) -> tuple[list[int], list[float]]:
    """Profile-guided sharing ratios (DESIGN.md R-solver-11): ms[i][j] =
    isolated time of request i at device fraction fracs[j].  Returns
    (weights, predicted slowdowns)."""
    k, nf = len(ms), len(fracs)
    fr = (f64 * max(nf, 1))(*fracs)
    flat = (f64 * max(k * nf, 1))(*[x for row in ms for x in row])
    w = (u32 * max(k, 1))()
    sp = (f64 * max(k, 1))()
    check(lib.accel_guided_weights(k, nf, fr, flat, scale, w, sp))
    return list(w)[:k], list(sp)[:k]


def accel_overlap(start: list[float], end: list[float]) -> float:
    k = len(start)
    o = f64()
    check(lib.accel_overlap((f64 * k)(*start), (f64 * k)(*end), k, C.byref(o)))
    return o.value

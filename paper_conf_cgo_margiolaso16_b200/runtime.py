"""Python face of the C ABI: one `Accel` context per device.

Marshalling only -- solving, dispatch and every tenant computation run in
libaccel.so (C++ host runtime + sm_100a kernels).
"""
from __future__ import annotations

import os

# Enough hardware work queues for concurrent tenant streams; must be set before
# the CUDA context exists (the default of 8 would serialise streams).
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")

from . import abi  # noqa: E402
from .jobs import Job  # noqa: E402


class Accel:
    def __init__(self, device: int = 0, mode: int = abi.MODE_SHARED, policy: int = abi.POLICY_STATIC,
                 verify: bool = False, caps: abi.accel_caps | None = None,
                 chunks: dict[str, int] | None = None):
        """chunks: per-kernel override of the VGs taken per dequeue (PAPER.md
        §6.4 adaptive scheduling; 1 = the paper's "naive" variant)."""
        self.device = device
        self.ctx = abi.accel_init(device, mode, policy, verify, caps)
        self.mode, self.policy, self.verify = mode, policy, verify
        self.kids: dict[str, int] = {}
        for name in abi.accel_builtin_names():
            desc = abi.accel_builtin_kernel(name)
            if chunks and name in chunks:
                desc.chunk = chunks[name]
            self.kids[name] = abi.accel_kernel_register(self.ctx, desc)

    def close(self):
        if self.ctx:
            abi.accel_finalize(self.ctx)
            self.ctx = None

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        self.close()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def set_mode(self, mode: int, policy: int | None = None):
        policy = self.policy if policy is None else policy
        abi.accel_set_mode(self.ctx, mode, policy)
        self.mode, self.policy = mode, policy

    def kernel_info(self, name: str) -> abi.accel_kernel_info:
        return abi.accel_kernel_info_get(self.ctx, self.kids[name])

    def submit(self, jobs: list[Job], tenants: list[int] | None = None, e2e: bool = False,
               weights: list[int] | None = None, launch_events: bool = False, trace: bool = False,
               linear_order: bool = False) -> list[int]:
        """Submit jobs as one group arriving together, in list order.
        trace: record every virtual group (vg_trace)."""
        tenants = list(range(len(jobs))) if tenants is None else tenants
        weights = [1] * len(jobs) if weights is None else weights
        fl = ((abi.REQ_LAUNCH_EVENTS if launch_events else 0) | (abi.REQ_TRACE if trace else 0) |
              (abi.REQ_LINEAR_ORDER if linear_order else 0))
        reqs = [j.request(self.kids, t, e2e, w, fl) for j, t, w in zip(jobs, tenants, weights)]
        # Job buffers (device inputs, tensor maps) were filled on torch's
        # stream; libaccel launches on its own non-blocking streams, which do
        # not order behind it.  Only torch's stream is waited on, never the
        # device (requests already running keep running).
        import torch
        torch.cuda.current_stream(self.device).synchronize()
        return abi.accel_submit_group(self.ctx, reqs)

    def sync(self, rid: int = abi.ACCEL_ALL):
        abi.accel_sync(self.ctx, rid)

    def epoch(self):
        abi.accel_epoch(self.ctx)

    def stats(self, rid: int) -> abi.accel_req_stats:
        return abi.accel_stats(self.ctx, rid)

    def launch_stats(self, rid: int, n: int) -> list[abi.accel_launch_stat]:
        return abi.accel_launch_stats(self.ctx, rid, n)

    def launch_times(self, rid: int, n: int) -> list[float]:
        return abi.accel_launch_times(self.ctx, rid, n)

    def vg_trace(self, rid: int):
        """Per-VG records (t_start_ns, t_end_ns, sm, cta) of a traced request."""
        return abi.accel_vg_trace(self.ctx, rid)

    def release(self, rid: int = abi.ACCEL_ALL):
        abi.accel_release(self.ctx, rid)

    def run(self, jobs: list[Job], e2e: bool = False, **kw) -> list[abi.accel_req_stats]:
        """Submit, wait, collect stats, release."""
        ids = self.submit(jobs, e2e=e2e, **kw)
        self.sync()
        st = [self.stats(i) for i in ids]
        self.release()
        return st

"""Pinned host<->device copy rate for one stencil volume (67 MB), CUDA events:
the e2e leg's copy floor.

    python scripts/pcie_copy.py
"""
import torch
n = 512 * 512 * 64
h = torch.ones(n, dtype=torch.float32).pin_memory()
d = torch.empty(n, dtype=torch.float32, device="cuda")
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
for what in ("h2d", "d2h"):
    for _ in range(3):
        (d.copy_(h, non_blocking=True) if what == "h2d" else h.copy_(d, non_blocking=True))
    torch.cuda.synchronize()
    e0.record()
    for _ in range(10):
        (d.copy_(h, non_blocking=True) if what == "h2d" else h.copy_(d, non_blocking=True))
    e1.record(); torch.cuda.synchronize()
    ms = e0.elapsed_time(e1) / 10
    print(f"{what} {4*n/1e6:.1f} MB pinned: {ms:.3f} ms = {4*n/ms/1e6:.1f} GB/s")

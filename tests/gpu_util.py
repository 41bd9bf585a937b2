"""Helpers for the GPU parity tests."""
import numpy as np

# BASELINE.json north star: "The fp32 tenants must match within 1e-4 relative
# error".  DESIGN.md R-tol-1: near-cancelling outputs make a pure
# relative test ill-posed, so the relative error is taken against
# max(|ref|, 1e-2 * max|ref|).
RTOL = 1e-4
FLOOR = 1e-2


def assert_close_fp32(got, ref, rtol=RTOL, floor=FLOOR, what=""):
    got = np.asarray(got, dtype=np.float64)
    ref = np.asarray(ref, dtype=np.float64)
    assert got.shape == ref.shape, (got.shape, ref.shape)
    scale = np.maximum(np.abs(ref), floor * (np.abs(ref).max() if ref.size else 0.0))
    scale = np.where(scale == 0, 1.0, scale)
    err = np.abs(got - ref) / scale
    bad = np.argwhere(err > rtol)
    assert bad.size == 0, (f"{what}: {len(bad)} of {ref.size} outside {rtol} "
                           f"(worst {err.max():.3g} at {np.unravel_index(err.argmax(), err.shape)})")
    return float(err.max()) if err.size else 0.0

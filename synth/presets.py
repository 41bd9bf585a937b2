"""Size presets per tenant.

`tiny`    -- unit/parity tests: the oracle finishes in well under a second, and
             the grids still span several virtual groups with a ragged tail.
`small`   -- Parboil-like sizes; BASELINE.json config 1 uses stencil 64^3 and
             histo 256K uint8.
`default` -- B200-scaled: each tenant's native grid covers >= ~2 waves at full
             occupancy and runs ~1-3 ms in isolation, so that one request can
             occupy the whole device ("a kernel
             execution request typically represents a computational range that
             is large enough to occupy all the accelerator resources").
"""
from __future__ import annotations

from . import gen

PRESETS: dict[str, dict[str, dict]] = {
    "mop": {
        "tiny": dict(n=256 * 37 + 0, block=256, nconst=11),
        "small": dict(n=1 << 20, block=256),
        "default": dict(n=1 << 26, block=256),
    },
    "stencil": {
        "tiny": dict(nx=70, ny=21, nz=19, sweeps=3),
        "small": dict(nx=64, ny=64, nz=64, sweeps=100),
        "default": dict(nx=512, ny=512, nz=64, sweeps=100),
    },
    "histo": {
        "tiny": dict(n=100_003, bins=256, iters=2, sample_bytes=1),
        "small": dict(n=1 << 18, bins=256, iters=20, sample_bytes=1),
        "default": dict(n=1 << 24, bins=16384, iters=100, sample_bytes=4),
    },
    "bfs": {
        "tiny": dict(nv=3000),
        "small": dict(nv=1 << 12),
        "default": dict(nv=1 << 20),
    },
    "cutcp": {
        "tiny": dict(box=16.0, cutoff=6.0, h=1.0),
        "small": dict(box=20.0),
        "default": dict(box=60.0),
    },
    "tpacf": {
        "tiny": dict(npts=300, nsets=3),
        "small": dict(npts=256 * 4, nsets=4),
        "default": dict(npts=4096, nsets=64),
    },
    "spmv": {
        "tiny": dict(grid=23, iters=2),
        "small": dict(grid=32, iters=100),
        "default": dict(grid=384, iters=100),
    },
    "sgemm": {
        "tiny": dict(m=200, n=136, k=72),
        "small": dict(m=1024, n=1056, k=992),
        "default": dict(m=4096, n=4096, k=4096),
    },
    "sad": {
        "tiny": dict(w=48, h=32, R=4),
        "small": dict(w=176, h=144, R=16),     # QCIF
        "default": dict(w=1920, h=1072, R=16),  # [ext Parboil sad large]
    },
    "histo_pipeline": {
        "tiny": dict(n=100_003, bins=16384, iters=2),
        "small": dict(n=1 << 18, bins=4096, iters=3),
        "default": dict(n=1 << 24, bins=16384, iters=20),
    },
    "gridding": {
        "tiny": dict(G=24, n=3000),
        "small": dict(G=48, n=40000),
        "default": dict(G=128, n=1 << 19),
    },
    "lbm": {
        "tiny": dict(nx=20, ny=11, nz=9, steps=3),
        "small": dict(nx=32, ny=32, nz=32, steps=5),
        "default": dict(nx=128, ny=128, nz=128, steps=20),   # ~2.1 M cells [ext; Parboil 120 x 120 x 150]
    },
    "mriq": {
        "tiny": dict(nvox_1d=12, numk=300),
        "small": dict(nvox_1d=32, numk=3072),
        "default": dict(nvox_1d=128, numk=2048),
    },
}


def preset(tenant: str, size: str = "default", seed: int = 0, **over) -> dict:
    """Generate the inputs of `tenant` at a named size (keyword overrides allowed)."""
    kw = dict(PRESETS[tenant][size])
    kw.update(over)
    return gen.GENERATORS[tenant](seed=seed, **kw)

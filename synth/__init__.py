"""Seeded synthetic inputs shared by the CPU oracle and the CUDA path.

This package holds ONLY input generation (random draws, data layout of the
inputs).  It contains none of the method's arithmetic: no share solving, no
dispatch, no tenant computation.  Both `oracle/` and the CUDA path consume the
arrays it returns; neither imports the other.

The workloads are shaped after the Parboil kernels the paper evaluates
(§7.2: "We use all the kernels from the OpenCL version
of the Parboil benchmark suite"); the paper only names them, so every shape
below is a synthetic [ext] recipe, stated in DESIGN.md §"Input recipe".
"""
from .gen import *  # noqa: F401,F403
from .presets import PRESETS, preset  # noqa: F401

"""B200-native accelOS hot path: fair space sharing of one GPU by concurrent
tenant kernels (Margiolas & O'Boyle, CGO'16).

libaccel.so (include/accel.h) holds the product: share solver, Virtual-NDRange
dispatch, native baseline, the tenant kernels.  `abi` is the ctypes binding
(same names as the C ABI), `jobs` builds tenant requests, `runtime.Accel` is a
convenience context.
"""
import os

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")

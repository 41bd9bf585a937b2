"""The C-ABI library loads on a CPU-only host and exports every entry point
include/accel.h declares (no compute calls without a GPU)."""
import ctypes
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _declared(header):
    txt = open(os.path.join(ROOT, "include", header)).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    return sorted(set(re.findall(r"\b(accel_[a-z_0-9]+)\s*\(", txt)))


def test_header_symbols_exported():
    from paper_conf_cgo_margiolaso16_b200 import abi
    names = _declared("accel.h")
    assert len(names) >= 20
    lib = ctypes.CDLL(abi.LIB_PATH)
    for n in names:
        assert hasattr(lib, n), n
    assert sorted(abi.EXPORTS) == names
    out = subprocess.check_output(["nm", "-D", "--defined-only", abi.LIB_PATH]).decode()
    for n in names:
        assert re.search(rf"\bT {n}\b", out), n


def test_builtins_listed():
    from paper_conf_cgo_margiolaso16_b200 import abi
    names = abi.accel_builtin_names()
    for n in ("mop", "stencil", "histo"):
        assert n in names
        d = abi.accel_builtin_kernel(n)
        assert d.persistent_fn and d.native_fn and d.persistent_fn != d.native_fn
        assert d.block.x in (128, 256) and d.args_size > 0
    with pytest.raises(abi.AccelError):
        abi.accel_builtin_kernel("nope")


def test_arg_struct_sizes_match_header():
    """ctypes mirrors vs the C compiler's view of include/accel_tenants.h."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    for n in abi.accel_builtin_names():
        d = abi.accel_builtin_kernel(n)
        cls = getattr(abi, f"accel_{n}_args")
        assert ctypes.sizeof(cls) == d.args_size, n


def test_struct_layouts_match_c(tmp_path):
    """sizeof of every ABI struct, from gcc, equals the ctypes mirror."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    structs = ["accel_dim3", "accel_caps", "accel_config", "accel_kernel_desc", "accel_kernel_info",
               "accel_launch", "accel_clear", "accel_copy", "accel_request", "accel_req_stats",
               "accel_demand", "accel_mix_metrics", "accel_mop_args", "accel_stencil_args",
               "accel_histo_args", "accel_bfs_args", "accel_cutcp_args", "accel_tpacf_args",
               "accel_spmv_args", "accel_sgemm_args", "accel_sgemm_split_args", "accel_sgemm_tc_args",
               "accel_mriq_phimag_args", "accel_mriq_q_args", "accel_stencil_tma_args", "accel_sad_args",
               "accel_lbm_args", "accel_histo_pre_args", "accel_gridding_args"]
    src = tmp_path / "s.c"
    src.write_text('#include <stdio.h>\n#include "accel.h"\n#include "accel_tenants.h"\nint main(){\n' +
                   "".join(f'printf("%zu\\n", sizeof({s}));\n' for s in structs) + "return 0;}\n")
    exe = tmp_path / "s"
    subprocess.check_call(["gcc", "-I", os.path.join(ROOT, "include"), str(src), "-o", str(exe)])
    sizes = [int(x) for x in subprocess.check_output([str(exe)]).split()]
    for s, n in zip(structs, sizes):
        assert ctypes.sizeof(getattr(abi, s)) == n, s


def test_init_without_gpu_fails_cleanly():
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    from paper_conf_cgo_margiolaso16_b200 import abi
    with pytest.raises(abi.AccelError) as e:
        abi.accel_init(0)
    assert e.value.code == abi.ACCEL_ECUDA


def test_pure_host_functions_validate():
    from paper_conf_cgo_margiolaso16_b200 import abi
    with pytest.raises(abi.AccelError) as e:
        abi.accel_demand_of(256, 32, 240 * 1024, 10)
    assert e.value.code == abi.ACCEL_ENOFIT
    with pytest.raises(abi.AccelError):
        abi.accel_metrics([1.0, 0.0], [1.0, 1.0])


def test_useful_occupancy_caps():
    """kMaxCtasPerSm reaches the descriptor (0 = no cap) -- values measured
    with scripts/occ_scaling.py, R-solver-10."""
    from paper_conf_cgo_margiolaso16_b200 import abi
    want = {"mriq_q": 1, "histo_wide": 0, "histo": 0, "bfs": 2, "spmv": 4, "tpacf": 3, "stencil": 0, "cutcp": 4}
    for n, v in want.items():
        assert abi.accel_builtin_kernel(n).max_ctas_per_sm == v, n

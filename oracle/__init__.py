"""CPU ORACLE -- TEST INFRASTRUCTURE ONLY.

Plain, slow, obviously-correct CPU implementations of everything the accelOS
hot path computes (PAPER.md = Margiolas & O'Boyle, CGO'16):

* `solver_ref`  -- the resource-sharing algorithm of §3 (PAPER.md 483-542),
                   step by step, with the readings of DESIGN.md §Readings.
* `metrics_ref` -- the fairness / throughput metrics of §7.4 (PAPER.md 877-913).
* `tenants`     -- liboracle (plain C, fp64 where the tenant is fp32, the
                   fp32 op sequence wherever a float decides an integer) for
                   the Fig. 8 `mop` kernel and the eight Parboil-shaped tenants.
* `dispatch_ref` -- the Virtual-NDRange dispatch semantics of Fig. 8b / §2.4
                   as a sequential simulation (coverage, decode, termination).

Only `tests/`, `__graft_entry__.smoke()` and `bench.py`'s cpu_baseline /
`--impl reference` legs may import or execute anything in this package.  It
shares no code with the CUDA path (`paper_conf_cgo_margiolaso16_b200/`), and
neither imports the other; both consume the seeded inputs of `synth/`.
"""

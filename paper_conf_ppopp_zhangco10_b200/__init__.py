"""B200-native batched tridiagonal solvers: CR, PCR, RD, CR+PCR, CR+RD
(Zhang, Cohen, Owens, "Fast Tridiagonal Solvers on the GPU", PPoPP'10).

The compute path is libtridiag.so (hand-written sm_100a CUDA behind the C ABI
of include/tridiag.h); this package is its ctypes binding plus the seeded
input generator (``inputs``) and the multi-GPU batch partitioner
(``partition``).
"""
from .tridiag import (ALGOS, HYBRIDS, TridiagError, abi_version, auto_switch_level,  # noqa: F401
                      host_workspace_bytes, last_kernel_names, last_launch_count, lib_path, load, max_n, phase_stamps,
                      max_switch_level, paper_cr, reload_knobs, solve_batched, solve_batched_host, solve_batched_raw,
                      solve_batched_strided_raw, solve_batched_large, large_workspace_bytes,
                      max_n_large, large_chunk, solve_batched_strided_large,
                      strided_large_workspace_bytes, column_chunk,
                      status_string)

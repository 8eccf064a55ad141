"""C-ABI of libtridiag.so: loads, exports every declared symbol, and validates
arguments on the host before touching CUDA (CPU only; no compute calls)."""
import ctypes
import os
import re

import pytest

import paper_conf_ppopp_zhangco10_b200 as td

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "tridiag.h")

F32, F64 = 0, 1
CR, PCR, RD, CR_PCR, CR_RD = range(5)
# fake, distinct, 256-B aligned "device" pointers: validation never dereferences
A, B, C, D, X = (0x10000000 * (i + 1) for i in range(5))


def declared_functions():
    src = open(HEADER).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(tridiag_[a-z_]+)\s*\(", src)))


def test_library_loads_and_exports_every_declared_symbol():
    L = td.load()
    names = declared_functions()
    assert "tridiag_solve_batched" in names and len(names) >= 9
    for name in names:
        assert hasattr(L, name), name
    assert td.abi_version() == 1


def solve(n=512, S=4, dtype=F32, algo=CR, m=0, a=A, b=B, c=C, d=D, x=X):
    return td.solve_batched_raw(a, b, c, d, x, n, S, dtype, algo, m, None)


def test_null_pointers():
    for kw in ("a", "b", "c", "d", "x"):
        assert solve(**{kw: 0}) == -1
        assert solve(S=0, **{kw: 0}) == 0       # empty batch: pointers unused
    assert solve(S=0, a=0, b=0, c=0, d=0, x=0, n=0) == -2


@pytest.mark.parametrize("n", [-4, 0])
def test_bad_n(n):
    assert solve(n=n) == -2


@pytest.mark.parametrize("n", [1, 3, 6, 100, 513, 8191])
def test_ragged_n_is_accepted(n):
    """n need not be a power of two (padded to the next one, NEXT f2); only
    validation is exercised here (S = 0: no launch)."""
    assert solve(n=n, S=0) == 0
    assert solve(n=n, S=0, algo=CR_PCR, m=2) == 0


def test_n_too_large():
    for dtype in (F32, F64):
        for algo in range(6):
            mx = td.max_n(dtype, algo)
            assert mx >= 256 and (mx & (mx - 1)) == 0
            assert solve(n=2 * mx, dtype=dtype, algo=algo) == -3
            assert solve(n=mx + 1, dtype=dtype, algo=algo) == -3   # pads to 2 mx
    assert td.max_n(F32, CR_PCR) == 8192 and td.max_n(F64, CR_PCR) == 4096
    assert td.max_n(F32, 5) == 512 and td.max_n(F64, 5) == 256   # rd_stone: one warp
    assert td.max_n(7, CR) == 0 and td.max_n(F32, 9) == 0


def test_bad_num_systems_dtype_algo():
    assert solve(S=-1) == -4
    assert solve(dtype=2) == -5
    assert solve(dtype=-1) == -5
    assert solve(algo=6) == -6
    assert solve(algo=-1) == -6


def test_switch_level_validation():
    for algo in (CR, PCR, RD, 5):
        assert solve(algo=algo, m=4) == -7
    for algo in (CR_PCR, CR_RD):
        assert solve(algo=algo, m=3) == -7
        assert solve(algo=algo, m=1) == -7
        assert solve(algo=algo, m=1024, n=512) == -7
        assert solve(algo=algo, m=-2) == -7
        assert solve(algo=algo, n=8192, m=8192) == -7   # inner capacity (fp32: 4096)
        assert td.max_switch_level(F32, algo, 8192) == 4096
        assert td.max_switch_level(F64, algo, 4096) == 2048
        for n in (2, 64, 512, 8192):
            m = td.auto_switch_level(n, F32, algo)
            assert 2 <= m <= n and (m & (m - 1)) == 0
    assert td.auto_switch_level(512, F32, CR) == 0


def test_overlap_rules():
    n, S = 512, 4
    nbytes = n * S * 4
    assert solve(x=A) == -8
    assert solve(x=B + 4) == -8
    assert solve(x=C - nbytes + 4) == -8
    assert solve(x=D + 8) == -8          # partial overlap with d
    assert solve(x=D, S=0) == 0          # exact in-place is allowed (S=0: no launch)
    assert solve(x=D + nbytes, S=0) == 0


def test_zero_systems_is_a_no_op():
    for algo in range(5):
        assert solve(S=0, algo=algo) == 0
    assert td.last_launch_count() == 0


def test_status_strings():
    for s in range(-9, 1):
        assert isinstance(td.status_string(s), str) and td.status_string(s)
    assert ">= 1" in td.status_string(-2)


def test_python_errors_are_loud():
    with pytest.raises(ValueError):
        td.tridiag.check(-2)
    with pytest.raises(td.TridiagError):
        td.tridiag.check(2)


def test_host_workspace_size():
    assert td.host_workspace_bytes(512, F32, 1000) == 3 * 4 * 1000 * 512 * 4
    assert td.host_workspace_bytes(512, F64, 0) > 0
    L = td.load()
    # workspace too small -> -9 before any CUDA call
    st = L.tridiag_solve_batched_host(A, B, C, D, X, 512, 4, F32, CR, 0, 0x1000, 16, 2)
    assert st == -9


def strided(n=512, S=4, es=1, ss=512, **kw):
    args = dict(a=A, b=B, c=C, d=D, x=X, dtype=F32, algo=CR, m=0)
    args.update(kw)
    return td.solve_batched_strided_raw(args["a"], args["b"], args["c"], args["d"], args["x"], n, S,
                                        es, ss, args["dtype"], args["algo"], args["m"], None)


def test_stride_validation():
    assert strided(es=0, S=0) == -10
    assert strided(ss=0, S=0) == -10
    assert strided(es=2, ss=2000, S=4) == -10      # neither stride is 1
    assert strided(es=1, ss=100, S=4) == -10       # rows overlap (ss < n)
    assert strided(es=3, ss=1, S=4, n=8) == -10    # columns overlap (es < S)
    assert strided(es=1, ss=512, S=0) == 0         # contiguous
    assert strided(es=1, ss=600, S=0) == 0         # pitched rows
    assert strided(es=8, ss=1, S=0, n=8) == 0      # interleaved
    assert td.status_string(-10).startswith("invalid strides")


def large(n, S=4, dtype=F32, algo=CR, m=0, bottom_n=0, ws=0x60000000, ws_bytes=1 << 40):
    return int(td.load().tridiag_solve_batched_large(A, B, C, D, X, n, S, dtype, algo, m, bottom_n,
                                                     ws, ws_bytes, None))


def test_large_n_capacity_and_workspace():
    """NEXT f2 (n > tridiag_max_n): CR-family up to 2^30; the
    workspace holds 4 arrays of n/R per reduction level plus the chunk-boundary
    heads (validation only, S = 0 or a bad argument: no launch)."""
    for dtype in (F32, F64):
        for algo in (CR, CR_PCR, CR_RD):
            assert td.max_n_large(dtype, algo) == 1 << 30
        for algo in (PCR, RD):
            assert td.max_n_large(dtype, algo) == td.max_n(dtype, algo)
    assert td.large_chunk(F32) == 4096 and td.large_chunk(F64) == 2048
    # fits on chip: no workspace
    assert td.large_workspace_bytes(8192, 10, F32, CR) == 0
    # n = 2^20 fp32: levels 2^20 -> 2^16 -> 2^12; the reduced arrays, 256-B aligned
    # (the chunk heads live in shared memory since round 2)
    S = 3
    exp = 0
    for nl in (1 << 20, 1 << 16):
        exp += 4 * (-(-S * (nl >> 4) * 4 // 256) * 256)
    assert td.large_workspace_bytes(1 << 20, S, F32, CR) == exp
    # hybrids stop reducing at m: CR+PCR m = 4096 at n = 16384 is one 2-level pass
    assert td.large_workspace_bytes(16384, 1, F32, CR_PCR, 4096) == 4 * 4096 * 4
    with pytest.raises(ValueError):
        td.large_workspace_bytes(1 << 31, 1, F32, CR)


def test_large_n_validation():
    assert large(1 << 20, S=0) == 0
    assert large(1 << 31, S=0) == -3                       # beyond tridiag_max_n_large
    assert large(16384, S=0, algo=PCR) == -3               # PCR / RD have no CR levels
    assert large(16384, S=0, algo=RD) == -3
    assert large(16384, S=0, bottom_n=1000) == -11         # not a power of two
    assert large(16384, S=0, bottom_n=1024) == -11         # below chunk / 2
    assert large(16384, S=0, bottom_n=16384) == -11        # above tridiag_max_n
    assert large(16384, S=0, bottom_n=2048) == 0
    assert large(16384, S=4, ws_bytes=16) == -9            # workspace too small
    assert large(16384, S=4, ws=0) == -9
    assert large(16384, S=0, algo=CR_PCR, m=8192) == -7    # m > max inner m
    assert large(16384, S=0, algo=CR_PCR, m=3) == -7
    assert td.status_string(-11).startswith("invalid bottom_n")


def strided_large(n, S=4, es=None, ss=1, dtype=F32, algo=CR, m=0, bottom_n=0, ws=0x60000000,
                  ws_bytes=1 << 40):
    es = max(S, 64) if es is None else es
    return int(td.load().tridiag_solve_batched_strided_large(A, B, C, D, X, n, S, es, ss, dtype,
                                                             algo, m, bottom_n, ws, ws_bytes, None))


def test_strided_large_workspace():
    """Column passes (ADI column sweep, NEXT f1 + f2): 4 interleaved arrays of
    n >> kin rows per pass level, 256-B aligned; rows (es = 1) are the large-n
    plan; PCR / RD and n <= 32 R need none (validation only).  The last pass
    writes the reduced systems as contiguous rows of the same size."""
    assert td.column_chunk(F32) == 128 and td.column_chunk(F64) == 64
    # fp32 4096 x 4096 columns: one pass 4096 -> 256
    assert td.strided_large_workspace_bytes(4096, 4096, 4096, 1, F32, CR_PCR) == 4 * 4096 * 256 * 4
    # fp64: one pass 4096 -> 512 (log2 R = 3 levels; the reduced rows are solved on chip)
    assert td.strided_large_workspace_bytes(4096, 4096, 4096, 1, F64, CR) == 4 * 4096 * 512 * 8
    # an explicit bottom_n below the first reduced size forces more passes
    assert td.strided_large_workspace_bytes(4096, 4096, 4096, 1, F64, CR, 0, 256) == \
        4 * 4096 * 512 * 8 + 4 * 4096 * 64 * 8
    # columns beyond tridiag_max_n: passes until <= tridiag_max_n (2^16 -> 4096)
    assert td.strided_large_workspace_bytes(1 << 16, 64, 64, 1, F32, CR) == 4 * 64 * 4096 * 4
    S = 3  # ragged S: 256-B alignment of each array
    assert td.strided_large_workspace_bytes(2048, S, S, 1, F32, CR) == 4 * (-(-S * 128 * 4 // 256) * 256)
    for algo in (PCR, RD):
        assert td.strided_large_workspace_bytes(2048, 40, 40, 1, F32, algo) == 0
    assert td.strided_large_workspace_bytes(512, 40, 40, 1, F32, CR) == 0          # on chip
    # m = 1024: one pass of one level, the row kernels run PCR on the 1024 survivors
    assert td.strided_large_workspace_bytes(2048, 40, 40, 1, F32, CR_PCR, 1024) == 4 * 40 * 1024 * 4
    assert td.strided_large_workspace_bytes(2048, 40, 40, 1, F32, CR_PCR, 2048) == 0  # m = n: no CR level
    # rows: the large-n plan (pitched rows allowed)
    assert td.strided_large_workspace_bytes(1 << 20, 3, 1, 1 << 20, F32, CR) == \
        td.large_workspace_bytes(1 << 20, 3, F32, CR)
    assert td.strided_large_workspace_bytes(8192, 3, 1, 8200, F32, CR) == 0
    with pytest.raises(ValueError):
        td.strided_large_workspace_bytes(4096, 40, 40, 1, F32, CR, 0, 1000)


def test_strided_large_validation():
    assert strided_large(4096, S=0) == 0
    assert strided_large(4096, S=40, ws=0) == -9                 # passes need a workspace
    assert strided_large(4096, S=40, ws_bytes=1024) == -9
    assert strided_large(4096, S=40, bottom_n=1000) == -11        # not a power of two
    assert strided_large(4096, S=40, bottom_n=32) == -11          # below column chunk / 2
    assert strided_large(4096, S=40, bottom_n=16384) == -11       # above tridiag_max_n
    assert strided_large(4096, S=0, bottom_n=64) == 0
    assert strided_large(1 << 15, S=0) == 0                       # beyond tridiag_max_n: passes
    assert strided_large(1 << 15, S=0, algo=PCR) == -3            # PCR has no CR levels
    assert strided_large(4096, S=40, es=40, ss=2) == -10          # neither stride 1
    assert strided_large(4096, S=0, algo=CR_PCR, m=3) == -7
    assert strided_large(4096, S=0, algo=CR_PCR, m=8192) == -7

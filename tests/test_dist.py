"""Multi-GPU batch partitioning, exercised on CPU with gloo (world size 2).

The solve path has no collective (systems are independent);
what must hold across ranks is: the shards tile the batch exactly, each rank's
counter-based inputs are the global batch's bytes, results solved per shard
equal results solved whole (oracle here; the GPU version is
test_gpu_parity.test_deterministic_and_partition_invariant), and the timing
reduction takes the max over ranks.
"""
import argparse
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from paper_conf_ppopp_zhangco10_b200 import inputs
from paper_conf_ppopp_zhangco10_b200.partition import (all_shards, reduce_max, reduce_sum,
                                                       shard_range)


@pytest.mark.parametrize("S", [0, 1, 7, 8, 1000, 1 << 20, 131071])
@pytest.mark.parametrize("W", [1, 2, 3, 4, 8])
def test_shards_tile_the_batch(S, W):
    sh = all_shards(S, W)
    assert sh[0].lo == 0 and sh[-1].hi == S
    for a, b in zip(sh, sh[1:]):
        assert a.hi == b.lo
    counts = [s.count for s in sh]
    assert max(counts) - min(counts) <= 1 and sum(counts) == S


def test_bad_partition_args():
    with pytest.raises(ValueError):
        shard_range(10, 0, 0)
    with pytest.raises(ValueError):
        shard_range(10, 2, 2)
    with pytest.raises(ValueError):
        shard_range(-1, 2, 0)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, S, n, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        import bench
        # strong scaling: the partitioner's shard; weak: rank * S
        args = argparse.Namespace(total_systems=S, systems=0)
        lo, cnt, total, scaling = bench.rank_workload(args, rank, world)
        a, b, c, d = inputs.generate("dd", cnt, n, torch.float64, s0=lo)
        x = oracle.thomas(*[t.numpy() for t in (a, b, c, d)])
        # gather every shard's solution on every rank (test only: the bench never does this)
        sizes = [None] * world
        dist.all_gather_object(sizes, (lo, cnt))
        xs = [None] * world
        dist.all_gather_object(xs, x)
        tmax = reduce_max(float(rank + 1))
        tsum = reduce_sum(float(cnt))
        wk = bench.rank_workload(argparse.Namespace(total_systems=0, systems=5), rank, world)
        q.put((rank, sizes, [np.asarray(v) for v in xs], tmax, tsum, total, scaling, wk))
    finally:
        dist.destroy_process_group()


def test_gloo_world2_partition_generation_and_reduction():
    world, S, n = 2, 37, 64
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, S, n, q)) for r in range(world)]
    for p in procs:
        p.start()
    out = [q.get(timeout=120) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    import oracle
    a, b, c, d = inputs.generate("dd", S, n, torch.float64)
    x_whole = oracle.thomas(*[t.numpy() for t in (a, b, c, d)])
    for rank, sizes, xs, tmax, tsum, total, scaling, wk in out:
        assert sizes == [(0, 18), (18, 19)]
        assert np.array_equal(np.concatenate(xs), x_whole)   # shard solves == whole solve
        assert tmax == 2.0 and tsum == S
        assert total == S and scaling == "strong"
        assert wk == (rank * 5, 5, 10, "weak")


def _scatter_worker(rank, world, port, s, n, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        from paper_conf_ppopp_zhangco10_b200.partition import scatter_solve_gather
        root = inputs.generate("dd", world * s, n, torch.float64) if rank == 0 else (None,) * 4

        def solve(a, b, c, d):
            return torch.from_numpy(oracle.thomas(*[t.numpy() for t in (a, b, c, d)]))

        x_full, x = scatter_solve_gather(root, (s, n), solve)
        q.put((rank, None if x_full is None else x_full.numpy(), x.numpy()))
    finally:
        dist.destroy_process_group()


def test_gloo_world2_scatter_solve_gather():
    """The NVLink "with transfer" analogue (NEXT f4): the root's batch is
    scattered in equal shards, solved per rank, gathered back -- the gathered x
    is the whole-batch solve, and each rank solved exactly its own rows."""
    world, s, n = 2, 9, 32
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_scatter_worker, args=(r, world, port, s, n, q)) for r in range(world)]
    for p in procs:
        p.start()
    out = sorted((q.get(timeout=120) for _ in range(world)), key=lambda o: o[0])
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    import oracle
    a, b, c, d = inputs.generate("dd", world * s, n, torch.float64)
    x_whole = oracle.thomas(*[t.numpy() for t in (a, b, c, d)])
    assert out[1][1] is None
    assert np.array_equal(out[0][1], x_whole)
    for rank, _, x in out:
        assert np.array_equal(x, x_whole[rank * s:(rank + 1) * s])

"""Multi-GPU batch partitioner.

The systems of a batch are independent, so W ranks split them
into contiguous ranges with no collective on the solve path: rank r owns
systems [floor(r*S/W), floor((r+1)*S/W)) -- sizes differ by at most one --
and generates / solves / stores only those ("owner computes").  The only
communication is after the timed region: max of the per-rank elapsed times
(and any error statistics) over NCCL.
"""
from __future__ import annotations

import os
from dataclasses import dataclass


@dataclass(frozen=True)
class Shard:
    rank: int
    world: int
    lo: int  # first global system index
    hi: int  # one past the last

    @property
    def count(self) -> int:
        return self.hi - self.lo


def shard_range(num_systems: int, world: int, rank: int) -> Shard:
    if world < 1 or not 0 <= rank < world:
        raise ValueError(f"bad rank {rank} of world {world}")
    if num_systems < 0:
        raise ValueError("num_systems must be >= 0")
    lo = (rank * num_systems) // world
    hi = ((rank + 1) * num_systems) // world
    return Shard(rank, world, lo, hi)


def all_shards(num_systems: int, world: int):
    return [shard_range(num_systems, world, r) for r in range(world)]


def dist_env():
    """(rank, local_rank, world) from the torchrun environment (1 process if absent)."""
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", str(rank)))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    return rank, local, world


def reduce_max(value: float, group=None) -> float:
    """Max of a per-rank scalar over all ranks (identity without a process group)."""
    import torch
    import torch.distributed as dist
    if not (dist.is_available() and dist.is_initialized()) or dist.get_world_size() == 1:
        return float(value)
    backend = dist.get_backend(group)
    dev = torch.device("cuda", torch.cuda.current_device()) if backend == "nccl" else torch.device("cpu")
    t = torch.tensor([float(value)], dtype=torch.float64, device=dev)
    dist.all_reduce(t, op=dist.ReduceOp.MAX, group=group)
    return float(t.item())


def reduce_sum(value: float, group=None) -> float:
    import torch
    import torch.distributed as dist
    if not (dist.is_available() and dist.is_initialized()) or dist.get_world_size() == 1:
        return float(value)
    backend = dist.get_backend(group)
    dev = torch.device("cuda", torch.cuda.current_device()) if backend == "nccl" else torch.device("cpu")
    t = torch.tensor([float(value)], dtype=torch.float64, device=dev)
    dist.all_reduce(t, op=dist.ReduceOp.SUM, group=group)
    return float(t.item())


def scatter_solve_gather(root_arrays, shard_shape, solve, root: int = 0, group=None, events=None):
    """The multi-GPU "with transfer" path (the NVLink
    analogue of the paper's PCIe column): the whole batch starts on
    ONE rank (`root`), which scatters equal contiguous shards of a, b, c, d to
    every rank (over NVLink / NVSwitch with NCCL), every rank solves its shard
    with `solve(a, b, c, d) -> x`, and the x shards are gathered back to the
    root.  This is the context row only: the bench's own multi-GPU number keeps
    each rank's inputs resident (owner computes, no collective on the solve
    path, 8(e)).

    root_arrays: (a, b, c, d), each (W * s, n) on the root (ignored elsewhere).
    shard_shape: (s, n), the per-rank shard (equal shards: dist.scatter).
    events: optional [e0, e1, e2, e3] CUDA events recorded on the current
    stream around scatter / solve / gather (device timing per phase).
    Returns (x_full on the root else None, this rank's x shard).
    """
    import torch
    import torch.distributed as dist
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    ref = root_arrays[0] if rank == root else None
    dtype = ref.dtype if ref is not None else None
    # dtype / device of the shards: the root's arrays; other ranks use the
    # process group's device (CUDA for NCCL) and agree on the dtype via the root
    obj = [str(dtype).replace("torch.", "") if rank == root else None]
    dist.broadcast_object_list(obj, src=root, group=group)
    dtype = getattr(torch, obj[0])
    backend = dist.get_backend(group)
    device = torch.device("cuda", torch.cuda.current_device()) if backend == "nccl" else torch.device("cpu")
    mark = (lambda i: events[i].record()) if events is not None else (lambda i: None)
    shards = [torch.empty(shard_shape, dtype=dtype, device=device) for _ in range(4)]
    mark(0)
    for arr, out in zip(root_arrays if rank == root else (None,) * 4, shards):
        parts = list(arr.chunk(world, dim=0)) if rank == root else None
        if parts is not None and any(p.shape != tuple(shard_shape) for p in parts):
            raise ValueError("scatter_solve_gather needs W equal shards of shape shard_shape")
        dist.scatter(out, parts, src=root, group=group)
    mark(1)
    x = solve(*shards)
    mark(2)
    if rank == root:
        x_full = torch.empty((world * shard_shape[0], shard_shape[1]), dtype=dtype, device=device)
        dist.gather(x, list(x_full.chunk(world, dim=0)), dst=root, group=group)
    else:
        x_full = None
        dist.gather(x, None, dst=root, group=group)
    mark(3)
    return x_full, x

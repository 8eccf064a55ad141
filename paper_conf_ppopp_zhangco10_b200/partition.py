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

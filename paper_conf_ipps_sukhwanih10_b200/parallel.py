"""Multi-GPU rotation sharding (production FTMap distributes rotations
across nodes; the paper's future multi-GPU plan).

Every (probe, rotation) unit is scored and filtered independently (the filter is per
rotation), so ranks take contiguous, equal blocks of the probe-major unit
space and no data-path exchange is needed until the very end, where ONE all-gather
(NCCL over NVLink on GPUs, gloo in the CPU tests) assembles the fixed-size pose blocks.
"""
from __future__ import annotations

from typing import Callable, Tuple

import torch
import torch.distributed as dist


def shard_range(n_units: int, rank: int, world: int) -> Tuple[int, int]:
    """Contiguous block of units owned by ``rank`` (sizes differ by at most one)."""
    if world < 1 or not 0 <= rank < world:
        raise ValueError("bad rank/world")
    return (n_units * rank) // world, (n_units * (rank + 1)) // world


def block_size(n_units: int, world: int) -> int:
    return -(-n_units // world)


def gather_poses(local: torch.Tensor, n_units: int, group=None) -> torch.Tensor:
    """All-gather per-rank pose blocks ``[U_r][k][4]`` int32 into ``[n_units][k][4]``.

    Blocks are padded to the common size ceil(n_units / world) so one
    ``all_gather_into_tensor`` (a single NCCL allgather) moves them; the padding is
    dropped afterwards.
    """
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    b, e = shard_range(n_units, rank, world)
    U = block_size(n_units, world)
    k = local.shape[1]
    if local.shape[0] != e - b:
        raise ValueError("local block size does not match this rank's shard")
    send = torch.full((U, k, 4), -1, dtype=torch.int32, device=local.device)
    send[: e - b] = local
    recv = torch.empty((world * U, k, 4), dtype=torch.int32, device=local.device)
    dist.all_gather_into_tensor(recv, send, group=group)
    parts = [recv[r * U: r * U + (shard_range(n_units, r, world)[1] - shard_range(n_units, r, world)[0])]
             for r in range(world)]
    return torch.cat(parts, dim=0)


def dock_sharded(dock_block: Callable[[int, int], torch.Tensor], n_units: int, group=None) -> torch.Tensor:
    """Run ``dock_block(begin, end) -> [end-begin][k][4] int32`` on this rank's shard and
    all-gather the result.  On GPUs ``dock_block`` is ``dock_probe_batch`` into a device
    buffer; the CPU tests plug in the oracle."""
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    b, e = shard_range(n_units, rank, world)
    return gather_poses(dock_block(b, e), n_units, group)


def dock_probe_sharded(ctx, probes, rot, k: int = 4, rho: int = 1, group=None) -> torch.Tensor:
    """Multi-GPU hot path: this rank docks its unit block with libdock into a device
    buffer, then one NCCL all-gather assembles every rank's poses on every rank."""
    from .dock import dock_probe_batch
    n_units = len(probes) * int(rot.shape[0])

    def block(b, e):
        out = torch.empty((e - b, k, 4), dtype=torch.int32, device=f"cuda:{ctx.device}")
        if e > b:
            dock_probe_batch(ctx, probes, rot, b, e, k, rho, out=out)
        return out

    return dock_sharded(block, n_units, group)

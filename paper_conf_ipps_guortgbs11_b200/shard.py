"""Frame sharding across GPUs.

ArrayOL treats time as an array dimension and the
downscaler never couples two frames or two channels, so the stream
partitions into contiguous frame blocks with NO data-path collective.  One
process per GPU; the only cross-GPU traffic is after the timed region: a MAX
all-reduce of the per-rank elapsed time and an all-gather of the per-frame u64
checksums (NCCL over NVLink on GPUs, gloo in the CPU tests).
"""
from __future__ import annotations

from typing import Optional, Tuple

import torch
import torch.distributed as dist


def weak_range(rank: int, world: int, frames_per_rank: int) -> Tuple[int, int]:
    """Weak scaling: every rank owns `frames_per_rank` frames; global indices are disjoint."""
    if not (0 <= rank < world) or frames_per_rank < 0:
        raise ValueError("bad rank/world/frames")
    return rank * frames_per_rank, frames_per_rank


def strong_range(rank: int, world: int, total_frames: int) -> Tuple[int, int]:
    """Strong scaling: `total_frames` split into `world` contiguous blocks (sizes differ by <= 1)."""
    if not (0 <= rank < world) or total_frames < 0:
        raise ValueError("bad rank/world/frames")
    base, extra = divmod(total_frames, world)
    start = rank * base + min(rank, extra)
    return start, base + (1 if rank < extra else 0)


def gather_results(checksums: torch.Tensor, elapsed_ms: float, group: Optional[dist.ProcessGroup] = None,
                   counts=None):
    """Collect (max elapsed over ranks, all checksums in global frame order).

    checksums: this rank's per-frame u64 checksums (uint64 or int64 tensor, on the
    backend's device).  counts: per-rank frame counts when ranks hold different
    numbers of frames (strong scaling); default = equal counts.
    Returns (max_elapsed_ms, int64 tensor of all checksums on the same device)."""
    cs = checksums.view(torch.int64) if checksums.dtype == torch.uint64 else checksums.to(torch.int64)
    t = torch.tensor([float(elapsed_ms)], dtype=torch.float64, device=cs.device)
    if not dist.is_initialized():   # single process: nothing to exchange
        return float(t.item()), cs.clone()
    world = dist.get_world_size(group)
    dist.all_reduce(t, op=dist.ReduceOp.MAX, group=group)
    if counts is None:
        out = torch.empty(world * cs.numel(), dtype=torch.int64, device=cs.device)
        dist.all_gather_into_tensor(out, cs.contiguous(), group=group)
        return float(t.item()), out
    # ragged: pad to the largest count, gather, then strip the padding
    n = max(counts)
    pad = torch.zeros(n, dtype=torch.int64, device=cs.device)
    pad[:cs.numel()] = cs
    out = torch.empty(world * n, dtype=torch.int64, device=cs.device)
    dist.all_gather_into_tensor(out, pad, group=group)
    parts = [out[r * n: r * n + counts[r]] for r in range(world)]
    return float(t.item()), torch.cat(parts)

"""One process per GPU: row-range sharding and the partial-aggregate exchange.

The table is split into contiguous row ranges [r*n/G, (r+1)*n/G) -- the Fig 3
control vector floor(i*G/n) one level above CTAs and threads (P:L241-250,
P:L264-266).  Each rank runs the fused fragment on its own range (no
data-path collective); the only exchange is one all-gather of the small
per-rank partials vector (<= 4096 groups x 9 slots x 16 B), after which
every rank merges in rank order with vd_merge_partials (exact 128-bit /
f64, deterministic) -- NCCL has no 128-bit reduction, so an all-reduce of
int64 would not be exact for Q1's sum_charge at SF100 (reading A17).

torch.distributed is plumbing here: process groups and the collective.  On
GPUs the backend is NCCL over NVLink/NVSwitch; the host logic is covered on
CPU with gloo (tests/test_dist_gloo.py).
"""
from __future__ import annotations

from typing import List, Sequence, Tuple

from . import vd


def shard_range(n_total: int, rank: int, world: int, align: int = 1) -> Tuple[int, int]:
    """Row range of `rank`: [floor(r*n/G), floor((r+1)*n/G)), boundaries rounded
    down to a multiple of `align` rows (the last rank takes the tail)."""
    if world < 1 or not 0 <= rank < world:
        raise ValueError("bad rank / world")

    def cut(r):
        if r >= world:
            return n_total
        c = (r * n_total) // world
        return c - c % align

    return cut(rank), cut(rank + 1)


def all_gather_partials(local, group=None) -> List[bytes]:
    """All-gather every rank's partials buffer (a uint8 tensor of
    vd.partials_bytes(plan) bytes) -> list of host byte strings in rank order."""
    import torch
    import torch.distributed as dist
    world = dist.get_world_size(group)
    nb = local.numel()
    gathered = torch.empty(nb * world, dtype=torch.uint8, device=local.device)
    dist.all_gather_into_tensor(gathered, local.contiguous(), group=group)
    host = gathered.cpu().numpy().tobytes()
    return [host[r * nb:(r + 1) * nb] for r in range(world)]


def merge(plan: vd.vd_pipeline, cols: Sequence[vd.vd_column], dims: Sequence[vd.vd_column],
          parts: Sequence[bytes], float_aggs: Sequence[bool] = ()):
    """Rank-order merge of per-rank partials + the Fig 11 compaction
    (vd_merge_partials, host): {group: [aggs..., rows]}."""
    return vd.merge_partials(plan, cols, dims, parts, float_aggs)


def exchange_and_merge(plan, cols, dims, local, group=None, float_aggs: Sequence[bool] = ()):
    """The cross-GPU step of the hierarchical fold: all-gather + host merge."""
    return merge(plan, cols, dims, all_gather_partials(local, group), float_aggs)


class DeviceExchange:
    """The cross-GPU step kept on the device (no host round trip): NCCL
    all_gather_into_tensor of every rank's partials into one buffer, then
    vd_merge_partials_device (one CTA: rank-order int128/f64 merge + Fig 11
    compaction) into a device vd_result -- both enqueued on the caller's
    stream, so the pair can be captured in a CUDA graph behind the pipeline
    launch.  world == 1 skips the collective (the merge is the compaction)."""

    def __init__(self, plan, cols, dims, local, world: int, group=None):
        import torch
        self.plan, self.cols, self.dims, self.local, self.world, self.group = plan, cols, dims, local, world, group
        nb = local.numel()
        self.gathered = (torch.empty(nb * world, dtype=torch.uint8, device=local.device) if world > 1 else local)
        self.result = vd.DeviceResult(plan, local.device)

    def step(self, stream=None):
        if self.world > 1:
            import torch.distributed as dist
            dist.all_gather_into_tensor(self.gathered, self.local, group=self.group)
        vd.merge_partials_device(self.plan, self.cols, self.dims, self.gathered, self.world, self.result, stream)
        return self.result

"""Multi-GPU plumbing of the hot path: one process per GPU,
points sharded across ranks, one all-reduce of the per-polygon partials.

COUNT and SUM are distributive and AVG is algebraic, so
each rank runs the whole query on its own point shard (its own canvas tiles,
polygons replicated) and the ranks combine only the n_poly-sized partial
vectors -- the paper's own out-of-core batching combines partial results the
same way.  AVG is finalised after the reduction.

torch.distributed provides the process group (NCCL over NVLink on B200s;
gloo for the CPU tests of this logic).
"""
from __future__ import annotations

import torch
import torch.distributed as dist

from . import rj


def shard_range(n: int, rank: int, world: int):
    """Contiguous index range [lo, hi) of rank's shard of n points."""
    lo = (n * rank) // world
    hi = (n * (rank + 1)) // world
    return lo, hi


def allreduce_partials(count: torch.Tensor, total: torch.Tensor | None = None, group=None):
    """Sum the per-polygon partials over all ranks, in place.

    count: uint64/int64 [n_poly]; total: float64 [n_poly] or None.  One
    collective: COUNT and SUM are packed into a single int64 buffer (the
    float64 sums are reduced in their own call only when present, because a
    sum of bit patterns is not a sum of values)."""
    c = count.view(torch.int64) if count.dtype == torch.uint64 else count
    dist.all_reduce(c, op=dist.ReduceOp.SUM, group=group)
    if total is not None:
        dist.all_reduce(total, op=dist.ReduceOp.SUM, group=group)
    return count, total


def query_sharded(R: "rj.RasterJoin", desc, d_count: torch.Tensor, d_sum: torch.Tensor, d_value: torch.Tensor,
                  group=None):
    """Partials on this rank's shard -> all-reduce -> finalise (all on device).

    The query and the finalisation run on the context's stream (rj_get_stream),
    the collective on torch's current stream; each waits for the other, so any
    stream choice at rj_create is safe."""
    rj.rj_query_device(R.ctx, desc, d_count, d_sum)
    ctx_stream = torch.cuda.ExternalStream(rj.rj_get_stream(R.ctx))
    cur = torch.cuda.current_stream()
    cur.wait_stream(ctx_stream)
    if dist.get_backend(group) == "gloo":
        # gloo stages device tensors through the host outside the stream order
        cur.synchronize()
    allreduce_partials(d_count, d_sum if desc.agg != 0 else None, group)
    ctx_stream.wait_stream(cur)
    rj.rj_finalize_device(R.ctx, desc.agg, d_count, d_sum, d_value)
    cur.wait_stream(ctx_stream)
    return d_value

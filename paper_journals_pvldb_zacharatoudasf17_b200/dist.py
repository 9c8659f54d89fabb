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
                  group=None, d_packed: torch.Tensor | None = None):
    """Partials on this rank's shard -> ONE all-reduce -> finalise (all on device).

    COUNT all-reduces the int64 counts; SUM/AVG first pack counts and sums
    into one binary64 buffer of 2 n_poly (rj_pack_partials; counts are exact
    in binary64 below 2^53) so a single collective combines both, then
    rj_finalize_packed unpacks and finalises.  librj's calls run on the
    context's stream (rj_get_stream), the collective on torch's current
    stream, each ordered after the other by stream waits -- including the
    caller's pending work on the output tensors -- so any stream choice at
    rj_create is safe."""
    ctx_stream = torch.cuda.ExternalStream(rj.rj_get_stream(R.ctx))
    cur = torch.cuda.current_stream()
    ctx_stream.wait_stream(cur)                  # caller's work on d_count / d_sum / d_value first
    rj.rj_query_device(R.ctx, desc, d_count, d_sum)
    gloo = dist.get_backend(group) == "gloo"
    if desc.agg == 0:
        cur.wait_stream(ctx_stream)
        if gloo:
            cur.synchronize()                    # gloo stages device tensors through the host
        c = d_count.view(torch.int64) if d_count.dtype == torch.uint64 else d_count
        dist.all_reduce(c, op=dist.ReduceOp.SUM, group=group)
        ctx_stream.wait_stream(cur)
        rj.rj_finalize_device(R.ctx, desc.agg, d_count, d_sum, d_value)
    else:
        n = d_count.numel()
        if d_packed is None or d_packed.numel() < 2 * n:
            d_packed = torch.empty(2 * n, dtype=torch.float64, device=d_count.device)
        rj.rj_pack_partials(R.ctx, d_count, d_sum, d_packed)
        cur.wait_stream(ctx_stream)
        if gloo:
            cur.synchronize()
        dist.all_reduce(d_packed[:2 * n], op=dist.ReduceOp.SUM, group=group)
        ctx_stream.wait_stream(cur)
        rj.rj_finalize_packed(R.ctx, desc.agg, d_packed, d_count, d_value)
    cur.wait_stream(ctx_stream)
    return d_value


# ---- spatially compact shards (second milestone) -----------
#
# Index-range shards of time-ordered input are spatially random: every rank
# then rasterises every polygon over the whole canvas, a fixed per-rank cost
# that caps strong scaling.  Exchanging the points once at load time into x
# strips of equal point count (splitters = x-quantiles of an all-gathered
# sample, one all_to_all per column over NVLink) lets each rank query only
# the pixel window of its strip (a viewport): its spans and pieces
# shrink by the world size.  Pixels on a strip border are seen by two ranks
# with disjoint points, and the per-polygon partials still just add
# (distributivity), so no pixel ownership is needed.

def strip_splitters(x: torch.Tensor, world: int, group=None, sample: int = 1 << 16, box=None,
                    poly_weight: float = 0.0) -> torch.Tensor:
    """world-1 increasing x splitters (float64, on x's device) giving strips
    of about equal cost over all ranks' points (see splitters_from_sample)."""
    n = x.numel()
    if n:
        idx = torch.linspace(0, n - 1, sample, device=x.device).round().long()
        s = x[idx].to(torch.float64)
    else:
        s = torch.full((sample,), float("nan"), dtype=torch.float64, device=x.device)
    parts = [torch.empty_like(s) for _ in range(world)]
    dist.all_gather(parts, s, group=group)
    return splitters_from_sample(torch.cat(parts), world, box, poly_weight)


def splitters_from_sample(allv: torch.Tensor, world: int, box=None, poly_weight: float = 0.0) -> torch.Tensor:
    """Splitters at the k/world quantiles (k = 1..world-1) of the strip cost
    (1 - w) * (share of the points) + w * (share of the domain width) over a
    sample of x (NaN ignored).  w = poly_weight = 0 balances points only; a
    rank's polygon pass grows with its strip's width (it rasterises the
    polygons of its window), so w ~ the polygon pass's share of a one-GPU
    query balances the two."""
    allv = torch.sort(allv[~torch.isnan(allv)].to(torch.float64)).values
    n = allv.numel()
    if n == 0:
        return torch.zeros(world - 1, dtype=torch.float64, device=allv.device)
    if poly_weight <= 0.0 or box is None:
        k = torch.arange(1, world, device=allv.device) * n // world
        return allv[k]
    w = float(poly_weight)
    cost = (1.0 - w) * torch.arange(1, n + 1, device=allv.device, dtype=torch.float64) / n + \
        w * ((allv - box[0]) / (box[2] - box[0])).clamp(0.0, 1.0)
    cost, _ = torch.cummax(cost, 0)
    q = torch.arange(1, world, device=allv.device, dtype=torch.float64) / world
    k = torch.searchsorted(cost, q).clamp(max=n - 1)
    return allv[k]


def strip_of(x: torch.Tensor, splitters: torch.Tensor) -> torch.Tensor:
    """Destination rank of every point: the number of splitters <= x (NaN
    coordinates go to the last rank and are dropped at load)."""
    d = torch.bucketize(x.to(torch.float64), splitters, right=True)
    return torch.where(torch.isnan(x), torch.full_like(d, splitters.numel()), d)


def exchange(columns, dest: torch.Tensor, world: int, group=None):
    """Send every point (all its columns) to rank dest[i]; returns this
    rank's received columns (grouped by source rank, input order kept)."""
    order = torch.argsort(dest, stable=True)
    send = torch.bincount(dest, minlength=world).to(torch.int64)
    recv = torch.empty_like(send)
    dist.all_to_all_single(recv, send, group=group)
    s_l, r_l = send.tolist(), recv.tolist()
    out = []
    for c in columns:
        o = torch.empty(sum(r_l), dtype=c.dtype, device=c.device)
        dist.all_to_all_single(o, c[order].contiguous(), r_l, s_l, group=group)
        out.append(o)
    return out


def strip_window(box, splitters, rank: int, world: int, desc):
    """Pixel window (c0, 0, c1, H) of the canvas desc resolves to, holding
    every point of rank's strip [split[rank-1], split[rank]) -- exact, through
    the C ABI's rj_resolve_window (reading Z20)."""
    sp = [float(v) for v in splitters.tolist()] if hasattr(splitters, "tolist") else list(splitters)
    lo = -float("inf") if rank == 0 else sp[rank - 1]
    hi = float("inf") if rank == world - 1 else sp[rank]
    return rj.rj_resolve_window(box, desc, (lo, -float("inf"), hi, float("inf")))


def spatial_shard(x, y, cols, world: int, group=None, box=None, poly_weight: float = 0.0):
    """Load-time exchange: (x, y, cols) of this rank's index range ->
    (x, y, cols, splitters) of its x strip."""
    sp = strip_splitters(x, world, group, box=box, poly_weight=poly_weight)
    dest = strip_of(x, sp)
    got = exchange([x, y, *cols], dest, world, group)
    return got[0], got[1], got[2:], sp

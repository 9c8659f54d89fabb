"""Multi-process (world_size 2, gloo, CPU) test of the sharding / all-reduce
plumbing of paper_journals_pvldb_zacharatoudasf17_b200.dist: each rank
computes oracle partials on its shard, the product's allreduce_partials
combines them, and the result equals the unsharded oracle (COUNT exact, SUM
to 1e-12 relative).  The CUDA query itself is covered by the gpu tests."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        from datagen import configs as C
        from paper_journals_pvldb_zacharatoudasf17_b200 import dist as rjdist

        n = 120_001
        pts = C.taxi(n, fare=True)
        lo, hi = rjdist.shard_range(n, rank, world)
        P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
        cnt, s, _ = oracle.query(P, pts["x"][lo:hi], pts["y"][lo:hi], cols=[pts["fare"][lo:hi]], agg_col=0,
                                 W=2048, H=2048, mode="accurate")
        tc = torch.from_numpy(cnt.astype(np.int64))
        ts = torch.from_numpy(s.copy())
        rjdist.allreduce_partials(tc, ts)
        if rank == 0:
            q.put((tc.numpy().copy(), ts.numpy().copy()))
    finally:
        dist.destroy_process_group()


def test_shards_allreduce_to_unsharded():
    import oracle
    from datagen import configs as C
    from paper_journals_pvldb_zacharatoudasf17_b200 import dist as rjdist

    assert [rjdist.shard_range(10, r, 3) for r in range(3)] == [(0, 3), (3, 6), (6, 10)]
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    got = q.get(timeout=300)
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    n = 120_001
    pts = C.taxi(n, fare=True)
    P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
    cnt, s, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["fare"]], agg_col=0, W=2048, H=2048, mode="accurate")
    assert np.array_equal(got[0], cnt.astype(np.int64))
    assert np.allclose(got[1], s, rtol=1e-12, atol=0)


def _spatial_worker(rank, world, port, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        from datagen import configs as C
        from paper_journals_pvldb_zacharatoudasf17_b200 import dist as rjdist

        n = 90_001
        pts = C.taxi(n, fare=True)
        lo, hi = rjdist.shard_range(n, rank, world)
        cols = [torch.from_numpy(pts["t"][lo:hi].copy()), torch.from_numpy(pts["fare"][lo:hi].copy())]
        x, y, cols, sp = rjdist.spatial_shard(torch.from_numpy(pts["x"][lo:hi].copy()),
                                              torch.from_numpy(pts["y"][lo:hi].copy()), cols, world)
        xs = x.numpy()
        # every point lands in its strip
        lo_x = -np.inf if rank == 0 else float(sp[rank - 1])
        hi_x = np.inf if rank == world - 1 else float(sp[rank])
        assert np.all((xs >= lo_x) & (xs < hi_x))
        W = 4096
        from paper_journals_pvldb_zacharatoudasf17_b200 import rj
        view = rjdist.strip_window(C.NYC_BOX, sp, rank, world, rj.make_desc(W=W, H=W))
        P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
        preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
        out = []
        for mode in ("bounded", "accurate"):
            # the window must hold every point of the strip: the windowed query
            # equals the unwindowed one on this rank's points
            c_w, s_w, _ = oracle.query(P, xs, y.numpy(), cols=[c.numpy() for c in cols], preds=preds,
                                       agg_col=1, W=W, H=W, mode=mode, view=view)
            c_a, _, _ = oracle.query(P, xs, y.numpy(), cols=[c.numpy() for c in cols], preds=preds,
                                     agg_col=1, W=W, H=W, mode=mode)
            assert np.array_equal(c_w, c_a)
            tc = torch.from_numpy(c_w.astype(np.int64))
            ts = torch.from_numpy(s_w.copy())
            rjdist.allreduce_partials(tc, ts)
            out.append((tc.numpy().copy(), ts.numpy().copy()))
        if rank == 0:
            q.put((out, len(xs), view))
        else:
            q.put((None, len(xs), view))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 3])
def test_spatial_shards_allreduce_to_unsharded(world):
    """x-strip shards by all_to_all + per-rank pixel windows
    give the unsharded result (COUNT exact, SUM to 1e-12) in both modes, with
    balanced strips."""
    import oracle
    from datagen import configs as C

    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_spatial_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = [q.get(timeout=300) for _ in range(world)]
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    out = next(r[0] for r in res if r[0] is not None)
    sizes = [r[1] for r in res]
    n = 90_001
    assert sum(sizes) == n
    assert max(sizes) - min(sizes) <= 0.05 * n / world        # x-quantile strips balance the points
    widths = sorted(r[2][2] - r[2][0] for r in res)
    assert widths[-1] < 4096                                   # windows are strips, not the canvas
    pts = C.taxi(n, fare=True)
    P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    for (gc, gs), mode in zip(out, ("bounded", "accurate")):
        cnt, s, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"], pts["fare"]], preds=preds, agg_col=1,
                                 W=4096, H=4096, mode=mode)
        assert np.array_equal(gc, cnt.astype(np.int64)), mode
        assert np.allclose(gs, s, rtol=1e-12, atol=0), mode


def test_splitters_from_sample_cost_rule():
    """poly_weight = 0: point quantiles; = 1: equal-width strips; between:
    monotone in the weight (wider sparse strips shrink)."""
    from paper_journals_pvldb_zacharatoudasf17_b200 import dist as rjdist

    g = torch.Generator().manual_seed(3)
    v = torch.rand(200_000, generator=g, dtype=torch.float64) ** 3 * 100.0
    box = (0.0, 0.0, 100.0, 50.0)
    q = rjdist.splitters_from_sample(v, 4)
    assert torch.allclose(q, torch.quantile(v, torch.tensor([0.25, 0.5, 0.75], dtype=torch.float64)), atol=0.05)
    e = rjdist.splitters_from_sample(v, 4, box, 1.0)
    assert torch.allclose(e, torch.tensor([25.0, 50.0, 75.0], dtype=torch.float64), atol=0.05)
    prev = q
    for w in (0.1, 0.3, 0.6, 0.9):
        s = rjdist.splitters_from_sample(v, 4, box, w)
        assert torch.all(s[1:] > s[:-1])
        assert torch.all(s >= prev - 1e-9)          # the skewed sample: splitters move right with w
        prev = s
    v2 = v.clone()
    v2[::7] = float("nan")
    assert torch.all(torch.isfinite(rjdist.splitters_from_sample(v2, 8, box, 0.2)))

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

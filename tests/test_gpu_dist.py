"""The multi-GPU query path on one GPU: two ranks (gloo process group, both
on cuda:0 -- NCCL cannot put two ranks on one device) each load a point
shard, compute device partials with rj_query_device, all-reduce them through
paper_journals_pvldb_zacharatoudasf17_b200.dist.query_sharded and finalise
on the device.  The result must equal the oracle on the whole point set
(COUNT exact, AVG to 1e-9)."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

pytestmark = pytest.mark.gpu


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


N = 300_001


def _worker(rank, world, port, q, spatial=False):
    try:
        _run(rank, world, port, q, spatial)
    except BaseException as e:          # report, do not hang the parent
        import traceback
        q.put(("error", rank, traceback.format_exc()))
        raise


def _run(rank, world, port, q, spatial=False):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from datagen import configs as C
        from paper_journals_pvldb_zacharatoudasf17_b200 import dist as rjdist
        from paper_journals_pvldb_zacharatoudasf17_b200 import rj

        torch.cuda.set_device(0)
        pts = C.taxi(N, fare=True)
        lo, hi = rjdist.shard_range(N, rank, world)
        stream = torch.cuda.current_stream()
        R = rj.RasterJoin(C.NYC_BOX, device=0, stream=stream.cuda_stream)
        x, y, cols = pts["x"][lo:hi], pts["y"][lo:hi], [pts["t"][lo:hi], pts["fare"][lo:hi]]
        view = None
        if spatial:
            # x strips by all_to_all, each rank queries its window
            tx, ty, tc, sp = rjdist.spatial_shard(torch.from_numpy(x.copy()), torch.from_numpy(y.copy()),
                                                  [torch.from_numpy(c.copy()) for c in cols], world)
            x, y, cols = tx.numpy(), ty.numpy(), [c.numpy() for c in tc]
            view = rjdist.strip_window(C.NYC_BOX, sp, rank, world, rj.make_desc(W=4096, H=4096))
        R.load_points(x, y, cols)
        R.load_polygons(C.array_polys("neighborhoods"))
        out = {}
        for mode in ("bounded", "accurate"):
            desc = rj.make_desc(agg="avg", agg_column=1, preds=[(0, ">=", C.T_2012[0])], W=4096, H=4096, mode=mode,
                                view=view)
            n = R.n_poly
            d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda")
            d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")
            d_val = torch.zeros(n, dtype=torch.float64, device="cuda")
            rjdist.query_sharded(R, desc, d_cnt, d_sum, d_val)
            torch.cuda.synchronize()
            out[mode] = (d_cnt.cpu().numpy(), d_val.cpu().numpy())
        R.close()
        if rank == 0:
            q.put(("ok", rank, out))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("spatial", [False, True])
def test_sharded_query_allreduce_on_one_gpu(spatial):
    if not torch.cuda.is_available():
        pytest.skip("needs a CUDA device")
    import oracle
    from datagen import configs as C

    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, q, spatial)) for r in range(2)]
    for p in procs:
        p.start()
    status, rank, got = q.get(timeout=600)
    assert status == "ok", f"rank {rank} failed:\n{got}"
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0, p.exitcode
    pts = C.taxi(N, fare=True)
    P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
    for mode in ("bounded", "accurate"):
        cnt, s, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"], pts["fare"]],
                                 preds=[(0, ">=", C.T_2012[0])], agg_col=1, W=4096, H=4096, mode=mode)
        gc, gv = got[mode]
        assert np.array_equal(gc.astype(np.uint64), cnt), mode
        ov = oracle.avg(cnt, s)
        both = np.isnan(gv) & np.isnan(ov)
        assert np.all(both | (np.abs(gv - ov) <= 1e-9 * np.abs(ov))), mode

import sys, os; sys.path.insert(0, os.getcwd())
import numpy as np, oracle
from datagen import configs as C
from paper_journals_pvldb_zacharatoudasf17_b200 import rj
N=300_001
pts = C.taxi(N, fare=True)
P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
for lo,hi in ((0,N),(0,150000),(150000,N)):
    R = rj.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"][lo:hi], pts["y"][lo:hi], [pts["t"][lo:hi], pts["fare"][lo:hi]])
    R.load_polygons(C.array_polys("neighborhoods"))
    oc, os_, _ = oracle.query(P, pts["x"][lo:hi], pts["y"][lo:hi], cols=[pts["t"][lo:hi], pts["fare"][lo:hi]], preds=[(0, ">=", C.T_2012[0])], agg_col=1, W=4096, H=4096, mode="accurate")
    for var in (-1, 1):
        R.set_option(rj.OPT_PASS, var)
        for agg in ("count","avg"):
            c, v = R.query(agg=agg, agg_column=1, preds=[(0, ">=", C.T_2012[0])], W=4096, H=4096, mode="accurate")
            d = np.nonzero(c != oc)[0]
            print(lo,hi,var,agg, "mismatch polys", len(d), "sum diff", int(c.sum()) - int(oc.sum()), d[:5], c[d[:5]], oc[d[:5]], R.stats()["n_boundary"])
    R.close()

import sys, os; sys.path.insert(0, os.getcwd())
import numpy as np
from datagen import configs as C
from paper_journals_pvldb_zacharatoudasf17_b200 import rj
import oracle
N = 300_001
pts = C.taxi(N, fare=True)
P = oracle.Polys(C.array_polys("neighborhoods"), C.NYC_BOX)
bad = 0
for lo, hi in ((0, 150000), (150000, N)):
    oc, _, _ = oracle.query(P, pts["x"][lo:hi], pts["y"][lo:hi], cols=[pts["t"][lo:hi], pts["fare"][lo:hi]],
                            preds=[(0, ">=", C.T_2012[0])], agg_col=1, W=4096, H=4096, mode="accurate")
    R = rj.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"][lo:hi], pts["y"][lo:hi], [pts["t"][lo:hi], pts["fare"][lo:hi]])
    R.load_polygons(C.array_polys("neighborhoods"))
    for it in range(40):
        mode = "bounded" if it % 3 == 0 else "accurate"
        c, v = R.query(agg="avg", agg_column=1, preds=[(0, ">=", C.T_2012[0])], W=4096, H=4096, mode=mode)
        if mode == "accurate" and not np.array_equal(c, oc):
            d = np.nonzero(c != oc)[0]
            bad += 1
            print("MISMATCH", lo, it, d[:8], c[d[:8]].astype(np.int64) - oc[d[:8]].astype(np.int64), R.stats()["n_boundary"])
print("bad", bad)

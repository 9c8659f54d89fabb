"""Golden fixtures (tests/golden/*.json): small examples whose expected values
were derived by hand from the paper's definitions, the derivation written out
line by line in the fixture next to its citations.  The paper prints no
per-polygon numbers (its Fig. 3/4/7 are figure-only), so these
hand-worked cases are the pins that do not come from a closed-form identity.

The oracle is checked against them on CPU; the CUDA path (through the C ABI)
against them on the GPU -- both sides reach the golden values independently.
"""
import glob
import json
import math
import os

import numpy as np
import pytest

import oracle
from datagen import polygons as PG

HERE = os.path.dirname(__file__)
FIXTURES = sorted(glob.glob(os.path.join(HERE, "golden", "*.json")))


def _load(path):
    g = json.load(open(path))
    polys = [[np.asarray(r, dtype=np.float64) for r in poly] for poly in g["polygons"]]
    pts = np.asarray(g["points"], dtype=np.float64)
    t = np.asarray(g["t"], dtype=np.int32)
    return g, PG.flatten(polys), pts[:, 0].copy(), pts[:, 1].copy(), t


def _cases(g):
    """(key, mode, preds) for every expected query result of a fixture."""
    for key, e in g["expected"].items():
        if "mode" in e:
            yield key, e["mode"], [tuple(p) for p in e.get("preds", [])]


def _check(g, key, cnt, s, avg=None):
    e = g["expected"][key]
    assert [int(c) for c in cnt] == e["count"], (key, cnt)
    assert [float(v) for v in s] == [float(v) for v in e["sum"]], (key, s)
    if avg is not None:
        for c, v, a in zip(e["count"], e["sum"], avg):
            assert (math.isnan(a) and c == 0) or a == v / c, (key, avg)


@pytest.mark.parametrize("path", FIXTURES, ids=os.path.basename)
def test_golden_oracle(path):
    g, flat, x, y, t = _load(path)
    P = oracle.Polys(flat, g["domain"])
    W, H = g["canvas"]
    for key, mode, preds in _cases(g):
        cnt, s, kept = oracle.query(P, x, y, cols=[t], preds=preds, agg_col=0, W=W, H=H, mode=mode)
        _check(g, key, cnt, s, oracle.avg(cnt, s))
        if not preds:
            assert kept == len(x) - g["n_out_of_domain"]
    if "interval" in g["expected"]:
        pc = oracle.pixel_counts(x, y, g["domain"], W=W, H=H)
        ep, em = oracle.error_interval(P, W, H, pc)
        assert ep.tolist() == g["expected"]["interval"]["eplus"]
        assert em.tolist() == g["expected"]["interval"]["eminus"]


@pytest.mark.gpu
@pytest.mark.parametrize("path", FIXTURES, ids=os.path.basename)
def test_golden_gpu(path):
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available():
        pytest.skip("needs a CUDA device")
    rjmod = pytest.importorskip("paper_journals_pvldb_zacharatoudasf17_b200.rj")
    g, flat, x, y, t = _load(path)
    R = rjmod.RasterJoin(tuple(g["domain"]))
    n_ood = R.load_points(x, y, [t])
    assert int(n_ood) == g["n_out_of_domain"]
    R.load_polygons(flat)
    W, H = g["canvas"]
    for key, mode, preds in _cases(g):
        cnt, s = R.query(agg="sum", agg_column=0, preds=preds, W=W, H=H, mode=mode)
        _, a = R.query(agg="avg", agg_column=0, preds=preds, W=W, H=H, mode=mode)
        _check(g, key, cnt, s, a)
    if "interval" in g["expected"]:
        cnt, _, ep, em = R.query_interval(agg="count", W=W, H=H)
        assert cnt.tolist() == g["expected"]["bounded"]["count"]
        assert ep.tolist() == g["expected"]["interval"]["eplus"]
        assert em.tolist() == g["expected"]["interval"]["eminus"]

"""C-ABI boundary checks that need no GPU: the library builds and loads,
exports every entry point include/rj.h declares, and its host-only logic
(S0 canvas resolution) follows the readings in DESIGN.md."""
import math
import os
import re

import numpy as np
import pytest

import oracle
from paper_journals_pvldb_zacharatoudasf17_b200 import _build, rj

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def L():
    _build.build()
    return rj.lib()


def header_functions():
    src = open(os.path.join(ROOT, "include", "rj.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(rj_[a-z_]+)\s*\(", src)))


def test_exports_every_declared_symbol(L):
    names = header_functions()
    assert len(names) >= 18
    for n in names:
        assert hasattr(L, n), n
    assert set(names) == set(rj.EXPORTS)


def test_version_and_status_strings(L):
    assert b"sm_100a" in L.rj_version()
    for code, name in rj.STATUS.items():
        assert L.rj_status_str(code).decode() == name


@pytest.mark.parametrize("eps,W", [(80, 1024), (40, 2048), (20, 4096), (10, 8192)])
def test_resolve_epsilon_nyc(L, eps, W):
    q = rj.make_desc(epsilon=eps)
    assert rj.rj_resolve_canvas_domain((0, 0, 57920, 57920), q) == (W, W)
    assert oracle.resolve(57920, 57920, eps) == (W, W)      # same reading on both sides


def test_resolve_us_and_errors(L):
    assert rj.rj_resolve_canvas_domain((0, 0, 4.6e6, 2.9e6), rj.make_desc(epsilon=1000.0)) == (6506, 4102)
    assert rj.rj_resolve_canvas_domain((0, 0, 1, 1), rj.make_desc(W=640, H=480)) == (640, 480)
    # reading Z21: up to 2^17 a side; eps = 1 m on NYC -> 81912 (as the oracle)
    assert rj.rj_resolve_canvas_domain((0, 0, 57920, 57920), rj.make_desc(epsilon=1.0)) == (81912, 81912)
    assert oracle.resolve(57920, 57920, 1.0) == (81912, 81912)
    assert rj.rj_resolve_canvas_domain((0, 0, 1, 1), rj.make_desc(W=131072)) == (131072, 131072)
    for q in (rj.make_desc(epsilon=0.0), rj.make_desc(epsilon=float("nan")), rj.make_desc(W=131073),
              rj.make_desc(epsilon=0.5)):    # eps = 0.5 m on NYC -> 163824 > 131072
        box = (0, 0, 57920, 57920)
        with pytest.raises(rj.RJError) as e:
            rj.rj_resolve_canvas_domain(box, q)
        assert e.value.status == -3


def test_create_without_gpu_fails_loudly(L):
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    with pytest.raises(rj.RJError) as e:
        rj.rj_create(0, None, (0, 0, 1, 1))
    assert e.value.status == -6


def test_create_rejects_bad_domain(L):
    for box in ((0, 0, 0, 1), (1, 0, 0, 1), (0, 0, math.inf, 1), (0, 0, 1, math.nan)):
        with pytest.raises(rj.RJError) as e:
            rj.rj_create(0, None, box)
        assert e.value.status == -1


def test_product_never_imports_oracle():
    pkg = os.path.join(ROOT, "paper_journals_pvldb_zacharatoudasf17_b200")
    for dp, _, fs in os.walk(pkg):
        for f in fs:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                s = open(os.path.join(dp, f)).read()
                assert "import oracle" not in s and "from oracle" not in s and "rj_oracle" not in s, f


def test_desc_layout_matches_header(L):
    # the ctypes mirror of rj_query_desc must match the C layout (view[4] last)
    import ctypes
    q = rj.make_desc(W=8, view=(1, 2, 3, 4))
    assert list(q.view) == [1, 2, 3, 4]
    # C layout: 3 x int32, 4 B padding, 5 x rj_pred (16 B), 2 x int32, double, mode, view[4], 4 B tail
    assert rj.rj_query_desc.pred.offset == 16 and rj.rj_query_desc.epsilon.offset == 104
    assert rj.rj_query_desc.view.offset == 116 and ctypes.sizeof(rj.rj_query_desc) == 136


def test_lod_view_helper():
    # zoom into [100, 150) x [100, 200) of [0,1024)^2 at 1000 px: an 20480-wide
    # virtual canvas and its window
    Wf, Hf, v = rj.lod_view((0, 0, 1024, 1024), (100, 100, 150, 200), 1000)
    assert (Wf, Hf) == (20480, 10240)
    assert v == (2000, 1000, 3000, 2000)


def test_resolve_window_exact_and_tight():
    """rj_resolve_window (reading Z20) against the oracle's O1/O2 maps: on
    random domains, canvases and world rectangles, every point of the
    half-open rectangle falls in the window, and the window is tight (its
    first and last columns/rows hold the rectangle's extreme points)."""
    import oracle
    rng = np.random.default_rng(99)
    for _ in range(300):
        x0, y0 = rng.uniform(-1e6, 1e6, 2)
        w, h = 10 ** rng.uniform(-3, 6, 2)
        box = (x0, y0, x0 + w, y0 + h)
        W, H = int(rng.integers(1, 131073)), int(rng.integers(1, 5000))
        q = rj.make_desc(W=W, H=H)
        a, b = np.sort(rng.uniform(x0 - 0.1 * w, x0 + 1.1 * w, 2))
        c, d = np.sort(rng.uniform(y0 - 0.1 * h, y0 + 1.1 * h, 2))
        if a == b or c == d:
            continue
        v = rj.rj_resolve_window(box, q, (a, c, b, d))
        assert 0 <= v[0] < v[2] <= W and 0 <= v[1] < v[3] <= H
        xs = np.concatenate([rng.uniform(a, b, 200), [a, np.nextafter(b, -np.inf)]])
        ys = np.concatenate([rng.uniform(c, d, 200), [c, np.nextafter(d, -np.inf)]])
        for vals, lo, hi, n, p0, p1 in ((xs, box[0], box[2], W, v[0], v[2]), (ys, box[1], box[3], H, v[1], v[3])):
            qv = np.array([oracle.quantize(float(t), lo, hi) for t in vals])
            inside = (qv >= 0) & (qv < (1 << 30))
            pix = (qv[inside] * n) >> 30
            assert np.all((pix >= p0) & (pix < p1))
            if inside[-2] and inside[-1]:
                assert pix.min() == p0 and pix.max() == p1 - 1
    # the whole domain and +-infinity
    q = rj.make_desc(W=777, H=555)
    assert rj.rj_resolve_window((0, 0, 1, 1), q, (-np.inf, -np.inf, np.inf, np.inf)) == (0, 0, 777, 555)
    with pytest.raises(rj.RJError):
        rj.rj_resolve_window((0, 0, 1, 1), q, (0.5, 0, 0.5, 1))

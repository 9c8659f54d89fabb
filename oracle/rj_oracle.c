/*
 * oracle/rj_oracle.c -- CPU ORACLE FOR RASTER JOIN.  TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs may load this library.  The product path
 * (paper_journals_pvldb_zacharatoudasf17_b200/, librj.so) never links,
 * imports or calls it; the two share no code, header, table or constant
 * generator -- only the SURVEY.md 8(c) definitions, restated here from the
 * paper.
 *
 * Plain, slow, obviously correct: every point is tested against every
 * polygon (only the polygon's half-open MBR is checked first, PAPER-silent
 * lemma L3: a point outside [xmin,xmax)x[ymin,ymax) fails the O3 test because
 * no edge can toggle it -- a bounding-box reject, no index, no blocking).
 * Floating point is binary64, compiled with -ffp-contract=off.
 *
 * Definitions (readings Z1-Z14 in DESIGN.md):
 *   O1  Q(x) = floor(((x - X0) / (X1 - X0)) * 2^30), binary64 RN, division.
 *       Points kept iff 0 <= Q < 2^30 on both axes; polygon vertices need
 *       0 <= Q <= 2^30.                               (transform: P:507-508)
 *   O2  pixel ix = (Qx * W) >> 30; centre cx(i) = ((2i+1) 2^29) / W (floor);
 *       pixel lattice extent [qlo(i), qhi(i)], qlo(i) = ceil(i 2^30 / W).
 *                                         (pixel-centre rule: P:561-562)
 *   O3  inside = even-odd PNPOLY over all rings, int64, half-open tie rule.
 *                                          ("ri contains p": P:722)
 *   O4  filters: conjunction, per-dtype compare.
 *   O5  bounded: every filtered point takes its pixel centre's membership.
 *                                           (Procs. DrawPoints/DrawPolygons,
 *                                            P:519-527, 4.2)
 *   O6  accurate: every filtered point takes its own membership.
 *                          (Procs. AccuratePoints/JoinPoint, 4.3)
 *   O7  AVG = SUM / COUNT, NaN when COUNT = 0.
 *   O8  COUNT uint64; SUM binary64 with Neumaier compensation.
 *   O9  boundary pixel: the segment meets the closed lattice rectangle of
 *       the pixel ("draw the outline", conservative raster P:880-887).
 *   O10 worst-case interval [A - e+, A + e-] over boundary pixels.
 *   O11 MIN / MAX (distributive; multiple aggregates P:1278-1283):
 *       the least / greatest attribute value of the polygon's points under
 *       IEEE 754 totalOrder for float32 (-NaN < -inf < ... < -0 < +0 < ...
 *       < +inf < +NaN, NaNs further ordered by payload; reading Z16), plain
 *       order for int32; NaN result for a polygon without points.
 *   O13 expected interval [A - E+, A + E-] with the pixel-polygon area
 *       fraction f (reading Z22).
 */
#include <math.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#ifdef _OPENMP
#include <omp.h>
#endif

#define OR_EXPORT __attribute__((visibility("default")))
#define OR_ONE30 ((int64_t)1 << 30)

/* ---------------------------------------------------------------- O1 / O2 */

/* O1: floor(((v - lo) / (hi - lo)) * 2^30) as int64; INT64_MIN for NaN or
 * values that do not fit (|.| >= 2^62). */
OR_EXPORT int64_t or_quantize(double v, double lo, double hi) {
    double d = v - lo;
    double s = hi - lo;
    double f = d / s;
    double g = f * 1073741824.0;           /* exact: power of two */
    double fl = floor(g);
    if (!(fl >= -4611686018427387904.0 && fl < 4611686018427387904.0)) return INT64_MIN;
    return (int64_t)fl;
}

/* O2 */
OR_EXPORT int64_t or_pixel(int64_t q, int64_t W) { return (q * W) >> 30; }
OR_EXPORT int64_t or_centre(int64_t i, int64_t W) { return ((2 * i + 1) * ((int64_t)1 << 29)) / W; }
static int64_t or_ceil_div_pos(int64_t a, int64_t b) { /* a >= 0, b > 0 */ return (a + b - 1) / b; }
OR_EXPORT int64_t or_qlo(int64_t i, int64_t W) { return or_ceil_div_pos(i * OR_ONE30, W); }
OR_EXPORT int64_t or_qhi(int64_t i, int64_t W) { return or_ceil_div_pos((i + 1) * OR_ONE30, W) - 1; }

/* S0 / reading Z3: epsilon -> resolution, W = ceil(w * sqrt(2) / eps).
 * Returns 0 on success, -1 for a bad epsilon or a resolution outside
 * [1, 131072] (reading Z21). */
#define OR_MAX_CANVAS 131072.0
OR_EXPORT int or_resolve(double w, double h, double eps, int *W, int *H) {
    if (!(eps > 0.0)) return -1;
    double a = ceil(w * sqrt(2.0) / eps);
    double b = ceil(h * sqrt(2.0) / eps);
    if (!(a >= 1.0 && a <= OR_MAX_CANVAS && b >= 1.0 && b <= OR_MAX_CANVAS)) return -1;
    *W = (int)a;
    *H = (int)b;
    return 0;
}

/* ---------------------------------------------------------------- polygons */

typedef struct {
    int64_t n_poly, n_ring, n_vert;
    int64_t *ring_off;   /* per polygon: first ring (n_poly+1) */
    int64_t *vert_off;   /* per ring: first vertex (n_ring+1) */
    int64_t *qx, *qy;    /* quantised vertices (O1) */
    int64_t *mbr;        /* per polygon: xmin, ymin, xmax, ymax (lattice) */
} or_polys;

/* Quantise the raw rings.  Returns NULL if a vertex is outside [0, 2^30]. */
OR_EXPORT or_polys *or_polys_new(int64_t n_poly, const uint32_t *poly_ring_off,
                                 const uint32_t *ring_vert_off, const double *vx,
                                 const double *vy, double x0, double y0, double x1, double y1) {
    or_polys *p = (or_polys *)calloc(1, sizeof(or_polys));
    p->n_poly = n_poly;
    p->n_ring = poly_ring_off[n_poly];
    p->n_vert = ring_vert_off[p->n_ring];
    p->ring_off = (int64_t *)malloc(sizeof(int64_t) * (n_poly + 1));
    p->vert_off = (int64_t *)malloc(sizeof(int64_t) * (p->n_ring + 1));
    p->qx = (int64_t *)malloc(sizeof(int64_t) * (p->n_vert + 1));
    p->qy = (int64_t *)malloc(sizeof(int64_t) * (p->n_vert + 1));
    p->mbr = (int64_t *)malloc(sizeof(int64_t) * 4 * (n_poly + 1));
    for (int64_t i = 0; i <= n_poly; ++i) p->ring_off[i] = poly_ring_off[i];
    for (int64_t i = 0; i <= p->n_ring; ++i) p->vert_off[i] = ring_vert_off[i];
    for (int64_t v = 0; v < p->n_vert; ++v) {
        p->qx[v] = or_quantize(vx[v], x0, x1);
        p->qy[v] = or_quantize(vy[v], y0, y1);
        if (p->qx[v] < 0 || p->qx[v] > OR_ONE30 || p->qy[v] < 0 || p->qy[v] > OR_ONE30) {
            free(p->ring_off); free(p->vert_off); free(p->qx); free(p->qy); free(p->mbr); free(p);
            return NULL;
        }
    }
    for (int64_t P = 0; P < n_poly; ++P) {
        int64_t xmin = INT64_MAX, ymin = INT64_MAX, xmax = INT64_MIN, ymax = INT64_MIN;
        for (int64_t r = p->ring_off[P]; r < p->ring_off[P + 1]; ++r)
            for (int64_t v = p->vert_off[r]; v < p->vert_off[r + 1]; ++v) {
                if (p->qx[v] < xmin) xmin = p->qx[v];
                if (p->qx[v] > xmax) xmax = p->qx[v];
                if (p->qy[v] < ymin) ymin = p->qy[v];
                if (p->qy[v] > ymax) ymax = p->qy[v];
            }
        p->mbr[4 * P + 0] = xmin; p->mbr[4 * P + 1] = ymin;
        p->mbr[4 * P + 2] = xmax; p->mbr[4 * P + 3] = ymax;
    }
    return p;
}

OR_EXPORT void or_polys_free(or_polys *p) {
    if (!p) return;
    free(p->ring_off); free(p->vert_off); free(p->qx); free(p->qy); free(p->mbr); free(p);
}

OR_EXPORT int64_t or_polys_vertex(const or_polys *p, int64_t v, int axis) {
    return axis == 0 ? p->qx[v] : p->qy[v];
}

/* O3: even-odd PNPOLY over every ring of polygon P (closing edge included).
 * Edge a->b toggles iff (ya > py) != (yb > py) and p lies strictly left of
 * the crossing: (px - xa)(yb - ya) < (xb - xa)(py - ya) for yb > ya, with the
 * inequality reversed for yb < ya.  Exact int64; |products| < 2^61. */
OR_EXPORT int or_pnpoly(const or_polys *p, int64_t P, int64_t px, int64_t py) {
    int inside = 0;
    for (int64_t r = p->ring_off[P]; r < p->ring_off[P + 1]; ++r) {
        int64_t v0 = p->vert_off[r], v1 = p->vert_off[r + 1];
        for (int64_t a = v0; a < v1; ++a) {
            int64_t b = (a + 1 < v1) ? a + 1 : v0;
            int64_t xa = p->qx[a], ya = p->qy[a], xb = p->qx[b], yb = p->qy[b];
            if ((ya > py) != (yb > py)) {
                int64_t lhs = (px - xa) * (yb - ya);
                int64_t rhs = (xb - xa) * (py - ya);
                if (yb > ya ? lhs < rhs : lhs > rhs) inside = !inside;
            }
        }
    }
    return inside;
}

/* O3 + lemma L3: MBR reject, then PNPOLY. */
static int or_contains(const or_polys *p, int64_t P, int64_t px, int64_t py) {
    const int64_t *m = p->mbr + 4 * P;
    if (px < m[0] || px >= m[2] || py < m[1] || py >= m[3]) return 0;
    return or_pnpoly(p, P, px, py);
}

/* --------------------------------------------------------------- O4 filter */
enum { OR_LT = 0, OR_LE = 1, OR_GT = 2, OR_GE = 3, OR_EQ = 4 };
enum { OR_I32 = 0, OR_F32 = 1, OR_F64 = 2 };

static int or_cmp_d(double a, int op, double b) {
    switch (op) {
    case OR_LT: return a < b;
    case OR_LE: return a <= b;
    case OR_GT: return a > b;
    case OR_GE: return a >= b;
    case OR_EQ: return a == b;
    }
    return 0;
}
static int or_cmp_f(float a, int op, float b) {
    switch (op) {
    case OR_LT: return a < b;
    case OR_LE: return a <= b;
    case OR_GT: return a > b;
    case OR_GE: return a >= b;
    case OR_EQ: return a == b;
    }
    return 0;
}

typedef struct {
    int n_cols;
    const void *const *cols;
    const int *dtypes;
    int n_pred;
    const int *pcol, *pop;
    const double *pval;
} or_filter;

/* O4: int32 columns compare exactly against the double constant; float32
 * columns compare in float32 against the constant cast to float32 (NaN fails). */
static int or_pass(const or_filter *f, size_t i) {
    for (int k = 0; k < f->n_pred; ++k) {
        int c = f->pcol[k];
        if (f->dtypes[c] == OR_I32) {
            int32_t v = ((const int32_t *)f->cols[c])[i];
            if (!or_cmp_d((double)v, f->pop[k], f->pval[k])) return 0;
        } else if (f->dtypes[c] == OR_F32) {
            float v = ((const float *)f->cols[c])[i];
            if (!or_cmp_f(v, f->pop[k], (float)f->pval[k])) return 0;
        } else {
            double v = ((const double *)f->cols[c])[i];
            if (!or_cmp_d(v, f->pop[k], f->pval[k])) return 0;
        }
    }
    return 1;
}

static double or_attr(const or_filter *f, int col, size_t i) {
    if (col < 0) return 1.0;
    if (f->dtypes[col] == OR_I32) return (double)((const int32_t *)f->cols[col])[i];
    if (f->dtypes[col] == OR_F32) return (double)((const float *)f->cols[col])[i];
    return ((const double *)f->cols[col])[i];
}

/* O1 for one point of the raw (f32 or f64) coordinate arrays; returns 0 if dropped */
static int or_point_q(const void *x, const void *y, int xy_f64, size_t i, double x0, double y0,
                      double x1, double y1, int64_t *qx, int64_t *qy) {
    double xv = xy_f64 ? ((const double *)x)[i] : (double)((const float *)x)[i];
    double yv = xy_f64 ? ((const double *)y)[i] : (double)((const float *)y)[i];
    *qx = or_quantize(xv, x0, x1);
    *qy = or_quantize(yv, y0, y1);
    return *qx >= 0 && *qx < OR_ONE30 && *qy >= 0 && *qy < OR_ONE30;
}

/* O12: is the pixel of lattice point (qx, qy) inside the window view =
 * {c0, r0, c1, r1} (half-open)?  NULL = the whole canvas. */
static int or_in_view(const int32_t *view, int64_t qx, int64_t qy, int W, int H) {
    if (!view) return 1;
    int64_t ix = or_pixel(qx, W), iy = or_pixel(qy, H);
    return ix >= view[0] && ix < view[2] && iy >= view[1] && iy < view[3];
}

/* Neumaier-compensated accumulate (O8) */
static inline void or_nadd(double *s, double *c, double v) {
    double t = *s + v;
    if (fabs(*s) >= fabs(v)) *c += (*s - t) + v;
    else *c += (v - t) + *s;
    *s = t;
}

/* ------------------------------------------------------------- O5/O6 query
 * mode 0 = bounded (O5: centre of the point's pixel), 1 = accurate (O6).
 * Outputs per polygon: cnt (uint64), sum (binary64, Neumaier); sum may be
 * NULL.  agg_col < 0 sums nothing.  nthreads <= 0: OpenMP default.
 * Returns the number of kept (in-domain) points that passed the filter. */
OR_EXPORT uint64_t or_query(const or_polys *p, uint64_t n, const void *x, const void *y, int xy_f64,
                            double x0, double y0, double x1, double y1,
                            int n_cols, const void *const *cols, const int *dtypes,
                            int agg_col, int n_pred, const int *pcol, const int *pop,
                            const double *pval, int W, int H, int mode, int nthreads,
                            uint64_t *cnt, double *sum, const int32_t *view) {
    or_filter f = {n_cols, cols, dtypes, n_pred, pcol, pop, pval};
    int64_t np = p->n_poly;
    uint64_t kept = 0;
#ifdef _OPENMP
    int nt = nthreads > 0 ? nthreads : omp_get_max_threads();
#else
    int nt = 1;
    (void)nthreads;
#endif
    uint64_t *tc = (uint64_t *)calloc((size_t)nt * np, sizeof(uint64_t));
    double *ts = (double *)calloc((size_t)nt * np, sizeof(double));
    double *tk = (double *)calloc((size_t)nt * np, sizeof(double));
    uint64_t *tkept = (uint64_t *)calloc((size_t)nt, sizeof(uint64_t));
    #pragma omp parallel num_threads(nt)
    {
#ifdef _OPENMP
        int tid = omp_get_thread_num();
#else
        int tid = 0;
#endif
        uint64_t *c = tc + (size_t)tid * np;
        double *s = ts + (size_t)tid * np;
        double *k = tk + (size_t)tid * np;
        #pragma omp for schedule(dynamic, 4096)
        for (long long ii = 0; ii < (long long)n; ++ii) {
            size_t i = (size_t)ii;
            int64_t qx, qy;
            if (!or_point_q(x, y, xy_f64, i, x0, y0, x1, y1, &qx, &qy)) continue;
            if (!or_pass(&f, i)) continue;
            if (!or_in_view(view, qx, qy, W, H)) continue;
            tkept[tid]++;
            int64_t px = qx, py = qy;
            if (mode == 0) {
                px = or_centre(or_pixel(qx, W), W);
                py = or_centre(or_pixel(qy, H), H);
            }
            double a = (sum && agg_col >= 0) ? or_attr(&f, agg_col, i) : 0.0;
            for (int64_t P = 0; P < np; ++P) {
                if (or_contains(p, P, px, py)) {
                    c[P] += 1;
                    if (sum && agg_col >= 0) or_nadd(&s[P], &k[P], a);
                }
            }
        }
    }
    for (int64_t P = 0; P < np; ++P) {
        uint64_t cc = 0;
        double ss = 0.0, kk = 0.0;
        for (int t = 0; t < nt; ++t) {
            cc += tc[(size_t)t * np + P];
            or_nadd(&ss, &kk, ts[(size_t)t * np + P]);
            or_nadd(&ss, &kk, tk[(size_t)t * np + P]);
        }
        cnt[P] = cc;
        if (sum) sum[P] = ss + kk;
    }
    for (int t = 0; t < nt; ++t) kept += tkept[t];
    free(tc); free(ts); free(tk); free(tkept);
    return kept;
}

/* O11: IEEE 754-2008 section 5.10 totalOrder(a, b) restricted to "a < b"
 * for binary32, written from the definition: numeric order first; equal
 * numbers are ordered by sign (-0 < +0); a NaN with the sign bit set is
 * below every number and a NaN without it above; two NaNs of one sign are
 * ordered by payload, larger payloads lying farther from zero. */
static int or_total_less_f32(float a, float b) {
    uint32_t ba, bb;
    memcpy(&ba, &a, 4);
    memcpy(&bb, &b, 4);
    const int sa = (ba >> 31) & 1, sb = (bb >> 31) & 1;
    const int na = isnan(a), nb = isnan(b);
    if (!na && !nb) {
        if (a < b) return 1;
        if (a > b) return 0;
        return sa && !sb;                        /* -0 < +0; equal otherwise */
    }
    if (na && nb) {
        if (sa != sb) return sa;                 /* -NaN < +NaN */
        const uint32_t pa = ba & 0x007FFFFFu, pb = bb & 0x007FFFFFu;
        return sa ? pa > pb : pa < pb;
    }
    if (na) return sa;                           /* -NaN below all, +NaN above all */
    return !sb;                                  /* b is NaN: a < +NaN, a > -NaN */
}

/* O11: per polygon MIN and MAX of attribute column agg_col (int32 or
 * float32) over the filtered points counted in the polygon under `mode`
 * (O5 / O6, as or_query).  mn / mx receive the value as binary64 (exact for
 * both dtypes), NaN for a polygon without points.  Sequential. */
OR_EXPORT void or_query_minmax(const or_polys *p, uint64_t n, const void *x, const void *y, int xy_f64,
                               double x0, double y0, double x1, double y1,
                               int n_cols, const void *const *cols, const int *dtypes,
                               int agg_col, int n_pred, const int *pcol, const int *pop,
                               const double *pval, int W, int H, int mode, double *mn, double *mx,
                               const int32_t *view) {
    or_filter f = {n_cols, cols, dtypes, n_pred, pcol, pop, pval};
    const int64_t np = p->n_poly;
    const int is_f32 = dtypes[agg_col] == OR_F32;
    uint8_t *seen = (uint8_t *)calloc((size_t)np, 1);
    int32_t *imn = (int32_t *)calloc((size_t)np, 4), *imx = (int32_t *)calloc((size_t)np, 4);
    float *fmn = (float *)calloc((size_t)np, 4), *fmx = (float *)calloc((size_t)np, 4);
    for (uint64_t i = 0; i < n; ++i) {
        int64_t qx, qy;
        if (!or_point_q(x, y, xy_f64, i, x0, y0, x1, y1, &qx, &qy)) continue;
        if (!or_pass(&f, i)) continue;
        if (!or_in_view(view, qx, qy, W, H)) continue;
        int64_t px = qx, py = qy;
        if (mode == 0) {
            px = or_centre(or_pixel(qx, W), W);
            py = or_centre(or_pixel(qy, H), H);
        }
        for (int64_t P = 0; P < np; ++P) {
            if (!or_contains(p, P, px, py)) continue;
            if (is_f32) {
                const float v = ((const float *)cols[agg_col])[i];
                if (!seen[P] || or_total_less_f32(v, fmn[P])) fmn[P] = v;
                if (!seen[P] || or_total_less_f32(fmx[P], v)) fmx[P] = v;
            } else {
                const int32_t v = ((const int32_t *)cols[agg_col])[i];
                if (!seen[P] || v < imn[P]) imn[P] = v;
                if (!seen[P] || v > imx[P]) imx[P] = v;
            }
            seen[P] = 1;
        }
    }
    for (int64_t P = 0; P < np; ++P) {
        mn[P] = !seen[P] ? NAN : is_f32 ? (double)fmn[P] : (double)imn[P];
        mx[P] = !seen[P] ? NAN : is_f32 ? (double)fmx[P] : (double)imx[P];
    }
    free(seen); free(imn); free(imx); free(fmn); free(fmx);
}

/* O7: AVG = SUM / COUNT, NaN for an empty polygon. */
OR_EXPORT void or_avg(int64_t n, const uint64_t *cnt, const double *sum, double *avg) {
    for (int64_t i = 0; i < n; ++i) avg[i] = cnt[i] ? sum[i] / (double)cnt[i] : NAN;
}

/* Per-point membership bitmask over the first 64 polygons, same rule as
 * or_query (filter applied: points failing it, or dropped by O1, get 0). */
OR_EXPORT void or_membership(const or_polys *p, uint64_t n, const void *x, const void *y, int xy_f64,
                             double x0, double y0, double x1, double y1,
                             int n_cols, const void *const *cols, const int *dtypes,
                             int n_pred, const int *pcol, const int *pop, const double *pval,
                             int W, int H, int mode, uint64_t *bits, const int32_t *view) {
    or_filter f = {n_cols, cols, dtypes, n_pred, pcol, pop, pval};
    int64_t np = p->n_poly < 64 ? p->n_poly : 64;
    #pragma omp parallel for schedule(dynamic, 1024)
    for (long long ii = 0; ii < (long long)n; ++ii) {
        size_t i = (size_t)ii;
        int64_t qx, qy;
        bits[i] = 0;
        if (!or_point_q(x, y, xy_f64, i, x0, y0, x1, y1, &qx, &qy)) continue;
        if (!or_pass(&f, i)) continue;
        if (!or_in_view(view, qx, qy, W, H)) continue;
        int64_t px = qx, py = qy;
        if (mode == 0) {
            px = or_centre(or_pixel(qx, W), W);
            py = or_centre(or_pixel(qy, H), H);
        }
        uint64_t m = 0;
        for (int64_t P = 0; P < np; ++P)
            if (or_contains(p, P, px, py)) m |= (uint64_t)1 << P;
        bits[i] = m;
    }
}

/* Pixel spans of one polygon from brute-force centre membership (O2 + O3,
 * pixel-centre rule P:561-562): every pixel centre of every row is tested
 * with O3, and maximal runs of inside centres are written as (row, lo, hi)
 * triples, hi exclusive; returns the count (or the required count if it
 * exceeds cap).  Pinned by tests/test_oracle_pins.py
 * test_pixel_spans_rectilinear_closed_form / _triangle_halfplanes. */
OR_EXPORT int64_t or_pixel_spans(const or_polys *p, int64_t P, int W, int H, int64_t cap, int32_t *out) {
    int64_t ns = 0;
    for (int r = 0; r < H; ++r) {
        int64_t cy = or_centre(r, H);
        int in = 0, lo = 0;
        for (int i = 0; i <= W; ++i) {
            int v = 0;
            if (i < W) v = or_contains(p, P, or_centre(i, W), cy);
            if (v && !in) { in = 1; lo = i; }
            else if (!v && in) {
                in = 0;
                if (ns < cap) { out[3 * ns] = r; out[3 * ns + 1] = lo; out[3 * ns + 2] = i; }
                ns++;
            }
        }
    }
    return ns;
}

/* ---------------------------------------------------------------------- O9
 * Does segment (xa,ya)-(xb,yb) meet the closed rectangle [x0,x1]x[y0,y1]?
 * Closed-bbox overlap, and not all four corner orientations of the same
 * strict sign (separating-axis test on the segment's line). */
static int or_orient(int64_t xa, int64_t ya, int64_t xb, int64_t yb, int64_t px, int64_t py) {
    int64_t v = (xb - xa) * (py - ya) - (yb - ya) * (px - xa);
    return (v > 0) - (v < 0);
}
OR_EXPORT int or_seg_rect(int64_t xa, int64_t ya, int64_t xb, int64_t yb,
                          int64_t x0, int64_t y0, int64_t x1, int64_t y1) {
    int64_t sx0 = xa < xb ? xa : xb, sx1 = xa < xb ? xb : xa;
    int64_t sy0 = ya < yb ? ya : yb, sy1 = ya < yb ? yb : ya;
    if (sx1 < x0 || sx0 > x1 || sy1 < y0 || sy0 > y1) return 0;
    int o1 = or_orient(xa, ya, xb, yb, x0, y0);
    int o2 = or_orient(xa, ya, xb, yb, x1, y0);
    int o3 = or_orient(xa, ya, xb, yb, x0, y1);
    int o4 = or_orient(xa, ya, xb, yb, x1, y1);
    if (o1 > 0 && o2 > 0 && o3 > 0 && o4 > 0) return 0;
    if (o1 < 0 && o2 < 0 && o3 < 0 && o4 < 0) return 0;
    return 1;
}

/* O9 boundary set B as a bitmask bits[r * ceil(W/32) + i/32] (union over the
 * polygons P in [p0, p1)).  Pixel extents exclude coordinate 2^30 (points
 * live in [0, 2^30)).  For each edge only the pixels inside the edge's
 * bounding box are visited; the others fail the bbox clause of O9. */
OR_EXPORT void or_boundary_mask(const or_polys *p, int64_t p0, int64_t p1, int W, int H, uint32_t *bits) {
    int64_t wpr = (W + 31) / 32;
    memset(bits, 0, sizeof(uint32_t) * (size_t)wpr * H);
    for (int64_t P = p0; P < p1; ++P)
        for (int64_t r = p->ring_off[P]; r < p->ring_off[P + 1]; ++r) {
            int64_t v0 = p->vert_off[r], v1 = p->vert_off[r + 1];
            for (int64_t a = v0; a < v1; ++a) {
                int64_t b = (a + 1 < v1) ? a + 1 : v0;
                int64_t xa = p->qx[a], ya = p->qy[a], xb = p->qx[b], yb = p->qy[b];
                int64_t sx0 = xa < xb ? xa : xb, sx1 = xa < xb ? xb : xa;
                int64_t sy0 = ya < yb ? ya : yb, sy1 = ya < yb ? yb : ya;
                if (sx0 >= OR_ONE30 || sy0 >= OR_ONE30) continue;
                if (sx1 > OR_ONE30 - 1) sx1 = OR_ONE30 - 1;
                if (sy1 > OR_ONE30 - 1) sy1 = OR_ONE30 - 1;
                int64_t i0 = or_pixel(sx0, W), i1 = or_pixel(sx1, W);
                int64_t r0 = or_pixel(sy0, H), r1 = or_pixel(sy1, H);
                for (int64_t rr = r0; rr <= r1; ++rr)
                    for (int64_t ii = i0; ii <= i1; ++ii) {
                        int64_t qx1 = or_qhi(ii, W), qy1 = or_qhi(rr, H);
                        if (qx1 > OR_ONE30 - 1) qx1 = OR_ONE30 - 1;
                        if (qy1 > OR_ONE30 - 1) qy1 = OR_ONE30 - 1;
                        if (or_seg_rect(xa, ya, xb, yb, or_qlo(ii, W), or_qlo(rr, H), qx1, qy1))
                            bits[rr * wpr + ii / 32] |= (uint32_t)1 << (ii % 32);
                    }
            }
        }
}

/* Filtered point counts per pixel C(pixel) (for O10).  out[r*W + i]. */
OR_EXPORT void or_pixel_counts(uint64_t n, const void *x, const void *y, int xy_f64,
                               double x0, double y0, double x1, double y1,
                               int n_cols, const void *const *cols, const int *dtypes,
                               int n_pred, const int *pcol, const int *pop, const double *pval,
                               int W, int H, uint32_t *out) {
    or_filter f = {n_cols, cols, dtypes, n_pred, pcol, pop, pval};
    memset(out, 0, sizeof(uint32_t) * (size_t)W * H);
    for (uint64_t i = 0; i < n; ++i) {
        int64_t qx, qy;
        if (!or_point_q(x, y, xy_f64, i, x0, y0, x1, y1, &qx, &qy)) continue;
        if (!or_pass(&f, i)) continue;
        out[or_pixel(qy, H) * W + or_pixel(qx, W)] += 1;
    }
}

/* O10: per polygon P, e+ = sum of C over P's own boundary pixels whose
 * centre is in P, e- = over those whose centre is not. */
OR_EXPORT void or_error_interval(const or_polys *p, int W, int H, const uint32_t *pixel_counts,
                                 uint64_t *eplus, uint64_t *eminus) {
    int64_t wpr = (W + 31) / 32;
    uint32_t *bits = (uint32_t *)malloc(sizeof(uint32_t) * (size_t)wpr * H);
    for (int64_t P = 0; P < p->n_poly; ++P) {
        or_boundary_mask(p, P, P + 1, W, H, bits);
        uint64_t ep = 0, em = 0;
        for (int64_t r = 0; r < H; ++r)
            for (int64_t i = 0; i < W; ++i)
                if (bits[r * wpr + i / 32] >> (i % 32) & 1) {
                    uint32_t c = pixel_counts[r * W + i];
                    if (or_contains(p, P, or_centre(i, W), or_centre(r, H))) ep += c;
                    else em += c;
                }
        eplus[P] = ep;
        eminus[P] = em;
    }
    free(bits);
}

/* --------------------------------------------------------------------- O13
 * Expected result interval: under a uniform distribution of the
 * points inside each pixel, a boundary pixel (x,y) of polygon i holds
 * f_i(x,y) x Fpt(x,y) points that are really inside i, where f_i(x,y) is
 * "the fraction area of the pixel that intersects polygon i".
 * Reading Z22: the garbled formula writes f_i for both sums; the
 * expected number of false positives in a P+ pixel (centre inside, whole
 * pixel counted) is (1 - f) Fpt and of false negatives in a P- pixel is
 * f Fpt, so
 *     E+_i = sum over P+_i of (1 - f_i) Fpt,  E-_i = sum over P-_i of f_i Fpt,
 * and the expected interval is [A - E+, A + E-].
 *
 * The pixel's region is the half-open lattice rectangle
 * [qlo(i), qlo(i+1)) x [qlo(r), qlo(r+1)) (O2: a lattice point Q stands for
 * [Q, Q+1), and the pixel of Q changes exactly at qlo).  Even-odd area of
 * polygon i inside it: every ring is clipped to the rectangle
 * (Sutherland-Hodgman; the clip of a closed ring against a convex window
 * keeps its signed area) and its signed shoelace area is added with weight
 * sigma_r = orientation(ring) * (-1)^depth(ring), depth = number of the
 * polygon's other rings containing the ring's first vertex (O3).  This is
 * the even-odd area whenever the rings of a polygon neither cross
 * themselves nor each other; for other rings it is the winding-weighted
 * area (reading Z22).  f is clamped to [0, 1]. */
static int or_ring_contains(const or_polys *p, int64_t r, int64_t px, int64_t py) {
    int inside = 0;
    int64_t v0 = p->vert_off[r], v1 = p->vert_off[r + 1];
    for (int64_t a = v0; a < v1; ++a) {
        int64_t b = (a + 1 < v1) ? a + 1 : v0;
        int64_t xa = p->qx[a], ya = p->qy[a], xb = p->qx[b], yb = p->qy[b];
        if ((ya > py) != (yb > py)) {
            int64_t lhs = (px - xa) * (yb - ya);
            int64_t rhs = (xb - xa) * (py - ya);
            if (yb > ya ? lhs < rhs : lhs > rhs) inside = !inside;
        }
    }
    return inside;
}

OR_EXPORT int or_ring_sigma(const or_polys *p, int64_t P, int64_t r) {
    __int128 s = 0;                                    /* twice the signed area, exact */
    int64_t v0 = p->vert_off[r], v1 = p->vert_off[r + 1];
    for (int64_t a = v0; a < v1; ++a) {
        int64_t b = (a + 1 < v1) ? a + 1 : v0;
        s += (__int128)p->qx[a] * p->qy[b] - (__int128)p->qx[b] * p->qy[a];
    }
    int orient = (s > 0) - (s < 0);
    int depth = 0;
    for (int64_t o = p->ring_off[P]; o < p->ring_off[P + 1]; ++o)
        if (o != r && or_ring_contains(p, o, p->qx[v0], p->qy[v0])) ++depth;
    return (depth & 1) ? -orient : orient;
}

/* keep the part of polygon (xs, ys)[n] with s * (coord - c) >= 0 on axis ax */
static int64_t or_clip_half(const double *xs, const double *ys, int64_t n, int ax, double c, double s,
                            double *ox, double *oy) {
    int64_t m = 0;
    for (int64_t k = 0; k < n; ++k) {
        int64_t l = (k + 1 < n) ? k + 1 : 0;
        double ak = s * ((ax ? ys[k] : xs[k]) - c), al = s * ((ax ? ys[l] : xs[l]) - c);
        if (ak >= 0) { ox[m] = xs[k]; oy[m] = ys[k]; ++m; }
        if ((ak >= 0) != (al >= 0)) {                 /* the edge crosses the line */
            double t = ak / (ak - al);
            if (ax) { ox[m] = xs[k] + t * (xs[l] - xs[k]); oy[m] = c; }
            else { ox[m] = c; oy[m] = ys[k] + t * (ys[l] - ys[k]); }
            ++m;
        }
    }
    return m;
}

OR_EXPORT double or_area_fraction(const or_polys *p, int64_t P, int64_t i, int64_t r, int W, int H) {
    int64_t X0 = or_qlo(i, W), X1 = or_qlo(i + 1, W), Y0 = or_qlo(r, H), Y1 = or_qlo(r + 1, H);
    double w = (double)(X1 - X0), h = (double)(Y1 - Y0), area = 0.0;
    for (int64_t rg = p->ring_off[P]; rg < p->ring_off[P + 1]; ++rg) {
        int64_t v0 = p->vert_off[rg], n = p->vert_off[rg + 1] - v0, cap = 16 * n + 64;
        double *buf = (double *)malloc(sizeof(double) * 4 * (size_t)cap);
        double *ax = buf, *ay = buf + cap, *bx = buf + 2 * cap, *by = buf + 3 * cap;
        for (int64_t k = 0; k < n; ++k) {              /* pixel-local coordinates (exact) */
            ax[k] = (double)(p->qx[v0 + k] - X0);
            ay[k] = (double)(p->qy[v0 + k] - Y0);
        }
        int64_t m = or_clip_half(ax, ay, n, 0, 0.0, 1.0, bx, by);      /* x >= 0 */
        m = or_clip_half(bx, by, m, 0, w, -1.0, ax, ay);               /* x <= w */
        m = or_clip_half(ax, ay, m, 1, 0.0, 1.0, bx, by);              /* y >= 0 */
        m = or_clip_half(bx, by, m, 1, h, -1.0, ax, ay);               /* y <= h */
        double s = 0.0;
        for (int64_t k = 0; k < m; ++k) {
            int64_t l = (k + 1 < m) ? k + 1 : 0;
            s += ax[k] * ay[l] - ax[l] * ay[k];
        }
        area += or_ring_sigma(p, P, rg) * 0.5 * s;
        free(buf);
    }
    double f = area / (w * h);
    return f < 0.0 ? 0.0 : (f > 1.0 ? 1.0 : f);
}

/* O13: expected interval sums over the same boundary pixels as O10. */
OR_EXPORT void or_expected_interval(const or_polys *p, int W, int H, const uint32_t *pixel_counts,
                                    double *eplus, double *eminus) {
    int64_t wpr = (W + 31) / 32;
    uint32_t *bits = (uint32_t *)malloc(sizeof(uint32_t) * (size_t)wpr * H);
    for (int64_t P = 0; P < p->n_poly; ++P) {
        or_boundary_mask(p, P, P + 1, W, H, bits);
        double ep = 0.0, em = 0.0, cp = 0.0, cm = 0.0;
        for (int64_t r = 0; r < H; ++r)
            for (int64_t i = 0; i < W; ++i)
                if (bits[r * wpr + i / 32] >> (i % 32) & 1) {
                    uint32_t c = pixel_counts[r * W + i];
                    if (!c) continue;
                    double f = or_area_fraction(p, P, i, r, W, H);
                    if (or_contains(p, P, or_centre(i, W), or_centre(r, H))) or_nadd(&ep, &cp, (1.0 - f) * c);
                    else or_nadd(&em, &cm, f * c);
                }
        eplus[P] = ep + cp;
        eminus[P] = em + cm;
    }
    free(bits);
}

/*
 * datagen/gen_points.c -- seeded synthetic point generators shared by the
 * oracle side (tests, cpu_baseline) and the CUDA side (bench, tests).
 *
 * This module holds NONE of Raster Join's arithmetic: no quantisation, no
 * pixel map, no point-in-polygon test.  It only draws world-coordinate
 * points and raw attribute columns, as a pure function of (seed, index), so
 * the output is identical for any thread count and any chunking (SURVEY.md
 * 8(d) "Seeds and generation").
 *
 * Workload shapes:
 *   uniform  -- C1: uniform f64 points in a box.
 *   taxi     -- C2/C3/C5: NYC-taxi-shaped mixture on a 57,920 m square
 *               (skew per PAPER.md P:1000-1003), t = seconds since 2009-01-01
 *               over 5 years, fare = cents-rounded log-normal.
 *   twitter  -- C4: 60 Zipf(1)-weighted city Gaussians + 15 % uniform on a
 *               4,600 x 2,900 km box, fav = geometric(p = 0.5).
 *
 * RNG: counter-based splitmix64 of (seed, stream, index); Box-Muller normals.
 */
#include <math.h>
#include <stdint.h>
#include <stddef.h>

#define DG_EXPORT __attribute__((visibility("default")))

static inline uint64_t dg_mix(uint64_t z) {
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ULL;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBULL;
    return z ^ (z >> 31);
}

/* One 64-bit draw for (seed, stream, index). */
DG_EXPORT uint64_t dg_u64(uint64_t seed, uint64_t stream, uint64_t index) {
    uint64_t z = seed * 0x9E3779B97F4A7C15ULL + stream * 0xD1B54A32D192ED03ULL +
                 index * 0xC2B2AE3D27D4EB4FULL + 0x632BE59BD9B4E019ULL;
    return dg_mix(dg_mix(z) + stream);
}

/* uniform in [0, 1) with 53 random bits */
static inline double dg_unif(uint64_t seed, uint64_t stream, uint64_t index) {
    return (double)(dg_u64(seed, stream, index) >> 11) * (1.0 / 9007199254740992.0);
}

/* a standard normal pair (Box-Muller) from streams s, s+1 */
static inline void dg_normal2(uint64_t seed, uint64_t s, uint64_t index, double *a, double *b) {
    double u1 = 1.0 - dg_unif(seed, s, index);     /* (0, 1] */
    double u2 = dg_unif(seed, s + 1, index);
    double r = sqrt(-2.0 * log(u1));
    double th = 6.283185307179586476925286766559 * u2;
    *a = r * cos(th);
    *b = r * sin(th);
}

static inline double dg_wrap(double v, double lo, double w) {
    double r = fmod(v - lo, w);
    if (r < 0) r += w;
    return lo + r;
}

/* ------------------------------------------------------------------ uniform */
DG_EXPORT void dg_uniform_points(uint64_t seed, uint64_t i0, uint64_t n,
                                 double x0, double y0, double x1, double y1,
                                 double *x, double *y) {
    #pragma omp parallel for schedule(static)
    for (long long k = 0; k < (long long)n; ++k) {
        uint64_t i = i0 + (uint64_t)k;
        x[k] = x0 + (x1 - x0) * dg_unif(seed, 0, i);
        y[k] = y0 + (y1 - y0) * dg_unif(seed, 1, i);
        if (x[k] >= x1) x[k] = x0;   /* guard the (measure-zero) rounding up to x1 */
        if (y[k] >= y1) y[k] = y0;
    }
}

/* --------------------------------------------------------------------- taxi */
/* Domain [0, 57920) x [0, 57920) metres (NYC-like). */
#define TAXI_W 57920.0
#define TAXI_T_SPAN 157766400      /* 5 years of seconds, 2009-01-01 .. 2013-12-31 */

DG_EXPORT void dg_taxi_points(uint64_t seed, uint64_t i0, uint64_t n,
                              float *x, float *y, int32_t *t, float *fare) {
    /* Manhattan-like axis: 29 degrees east of north */
    const double ang = (90.0 - 29.0) * 3.14159265358979323846 / 180.0;
    const double ux = cos(ang), uy = sin(ang);     /* major axis */
    const double vx = -uy, vy = ux;                /* minor axis */
    #pragma omp parallel for schedule(static)
    for (long long k = 0; k < (long long)n; ++k) {
        uint64_t i = i0 + (uint64_t)k;
        double c = dg_unif(seed, 0, i);
        double a, b;
        dg_normal2(seed, 1, i, &a, &b);
        double px, py;
        if (c < 0.65) {            /* elongated "Manhattan" Gaussian 4.5 km x 0.9 km */
            px = 24000.0 + a * 4500.0 * ux + b * 900.0 * vx;
            py = 33000.0 + a * 4500.0 * uy + b * 900.0 * vy;
        } else if (c < 0.75) {     /* "Midtown" hotspot, sigma 0.6 km */
            px = 24000.0 + 2000.0 * ux + a * 600.0;
            py = 33000.0 + 2000.0 * uy + b * 600.0;
        } else if (c < 0.81) {     /* airport 1, sigma 0.4 km */
            px = 36500.0 + a * 400.0;
            py = 17500.0 + b * 400.0;
        } else if (c < 0.85) {     /* airport 2, sigma 0.3 km */
            px = 32500.0 + a * 300.0;
            py = 36500.0 + b * 300.0;
        } else {                   /* broad background, sigma 8 km */
            px = 28960.0 + a * 8000.0;
            py = 28960.0 + b * 8000.0;
        }
        px = dg_wrap(px, 0.0, TAXI_W);
        py = dg_wrap(py, 0.0, TAXI_W);
        if (x) x[k] = (float)px;
        if (y) y[k] = (float)py;
        if (t) t[k] = (int32_t)(dg_u64(seed, 3, i) % (uint64_t)TAXI_T_SPAN);
        if (fare) {
            double g, h;
            dg_normal2(seed, 4, i, &g, &h);
            double v = 2.5 + 2.0 * exp(0.7 + 0.7 * g);
            fare[k] = (float)(floor(v * 100.0 + 0.5) / 100.0);
        }
    }
}

/* ------------------------------------------------------------------ twitter */
#define TW_W 4600000.0
#define TW_H 2900000.0
#define TW_CITIES 60

DG_EXPORT void dg_twitter_points(uint64_t seed, uint64_t i0, uint64_t n,
                                 float *x, float *y, int32_t *fav) {
    double cx[TW_CITIES], cy[TW_CITIES], cs[TW_CITIES], cdf[TW_CITIES];
    double tot = 0.0;
    for (int k = 0; k < TW_CITIES; ++k) {      /* city table: pure function of seed */
        cx[k] = 100000.0 + (TW_W - 200000.0) * dg_unif(seed, 100, (uint64_t)k);
        cy[k] = 100000.0 + (TW_H - 200000.0) * dg_unif(seed, 101, (uint64_t)k);
        cs[k] = 5000.0 + 35000.0 * dg_unif(seed, 102, (uint64_t)k);
        tot += 1.0 / (double)(k + 1);           /* Zipf(1) weights */
        cdf[k] = tot;
    }
    for (int k = 0; k < TW_CITIES; ++k) cdf[k] /= tot;
    #pragma omp parallel for schedule(static)
    for (long long k = 0; k < (long long)n; ++k) {
        uint64_t i = i0 + (uint64_t)k;
        double c = dg_unif(seed, 0, i);
        double px, py;
        if (c < 0.15) {
            px = TW_W * dg_unif(seed, 1, i);
            py = TW_H * dg_unif(seed, 2, i);
        } else {
            double u = dg_unif(seed, 5, i);
            int lo = 0, hi = TW_CITIES - 1;     /* first city with cdf > u */
            while (lo < hi) { int m = (lo + hi) / 2; if (cdf[m] > u) hi = m; else lo = m + 1; }
            double a, b;
            dg_normal2(seed, 1, i, &a, &b);
            px = cx[lo] + a * cs[lo];
            py = cy[lo] + b * cs[lo];
        }
        px = dg_wrap(px, 0.0, TW_W);
        py = dg_wrap(py, 0.0, TW_H);
        if (x) x[k] = (float)px;
        if (y) y[k] = (float)py;
        if (fav) {
            double u = 1.0 - dg_unif(seed, 6, i);  /* (0,1] */
            fav[k] = (int32_t)floor(log(u) / log(0.5));
        }
    }
}

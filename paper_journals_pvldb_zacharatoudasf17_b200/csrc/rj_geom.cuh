// rj_geom.cuh -- exact integer geometry of the GPU path (lattice, pixels,
// scanline thresholds, supercover).  Independent of oracle/ (shares no
// code): both sides implement the definitions written in DESIGN.md
// ("Readings of the paper"), which restate PAPER.md P:507-508 (transform),
// P:561-562 (pixel-centre rule), P:672-680/P:880-887 (boundary pixels).
//
// Lattice: 2^30 units per axis (k = 30).  Every intermediate below fits in
// signed 64-bit: |(x_b - x_a)(y - y_a)| < 2^60, x_a*den + dx*dy < 2^61,
// X*W <= 2^45.
#pragma once
#include <stdint.h>

#ifdef __CUDACC__
#define RJ_HD __host__ __device__ __forceinline__
#else
#define RJ_HD inline
#endif

namespace rj {

constexpr int kLatticeBits = 30;
constexpr int64_t kOne = int64_t(1) << kLatticeBits;      // 2^30
constexpr int64_t kHalf = int64_t(1) << (kLatticeBits - 1);
constexpr int kMaxLevel = 10;                              // finest point-cell level: 1024 x 1024
constexpr int kCells10 = 1 << (2 * kMaxLevel);             // cells at the finest level
constexpr int kGridBits = 10;                              // edge grid: 1024 x 1024
constexpr int kGrid = 1 << kGridBits;
constexpr int kGridShift = kLatticeBits - kGridBits;       // 20
constexpr int kMortonShift = kLatticeBits - 16;            // sort key: 16 bits per axis

// floor / ceil of a / 2^30 for signed a (arithmetic shift is floor)
RJ_HD int64_t floor_pow30(int64_t a) { return a >> kLatticeBits; }
RJ_HD int64_t ceil_pow30(int64_t a) { return -((-a) >> kLatticeBits); }
// floor / ceil of a / b for b > 0 (C '/' truncates toward zero)
RJ_HD int64_t ceil_div(int64_t a, int64_t b) {
    int64_t q = a / b, r = a - q * b;
    return q + (r > 0 ? 1 : 0);
}
RJ_HD int64_t floor_div(int64_t a, int64_t b) {
    int64_t q = a / b, r = a - q * b;
    return q - (r < 0 ? 1 : 0);
}
RJ_HD int64_t clamp64(int64_t v, int64_t lo, int64_t hi) { return v < lo ? lo : (v > hi ? hi : v); }

// pixel of a lattice coordinate q in [0, 2^30): (q*W) >> 30
RJ_HD int64_t pix(int64_t q, int64_t W) { return (q * W) >> kLatticeBits; }
// representative centre of pixel i: ((2i+1) 2^29) / W, inside pixel i
RJ_HD int64_t centre(int64_t i, int64_t W) { return ((2 * i + 1) * kHalf) / W; }
// first / last lattice coordinate of pixel i
RJ_HD int64_t qlo(int64_t i, int64_t W) { return ((i << kLatticeBits) + W - 1) / W; }
RJ_HD int64_t qhi(int64_t i, int64_t W) { return qlo(i + 1, W) - 1; }
// number of pixel rows whose centre lies below y: smallest r with centre(r) >= y
RJ_HD int64_t row_start(int64_t y, int64_t H) { return clamp64(ceil_pow30(y * H - kHalf), 0, H); }

// Scanline threshold of edge a->b (ya != yb) on pixel row r (its centre cy
// satisfies min(ya,yb) <= cy < max(ya,yb)): the edge toggles the even-odd
// membership of the centres of exactly the pixels i < t.
//   X* = xa + ceil((xb-xa)(cy-ya)/(yb-ya))  (smallest lattice x right of the crossing)
//   t  = clamp(ceil((X* W - 2^29) / 2^30), 0, W)
RJ_HD int64_t threshold(int64_t xa, int64_t ya, int64_t xb, int64_t yb, int64_t cy, int64_t W) {
    int64_t num = (xb - xa) * (cy - ya), den = yb - ya;
    if (den < 0) { num = -num; den = -den; }
    int64_t xs = xa + ceil_div(num, den);
    return clamp64(ceil_pow30(xs * W - kHalf), 0, W);
}

// Morton interleave of two 16-bit values (x in even bits)
RJ_HD uint32_t spread16(uint32_t v) {
    v &= 0xFFFFu;
    v = (v | (v << 8)) & 0x00FF00FFu;
    v = (v | (v << 4)) & 0x0F0F0F0Fu;
    v = (v | (v << 2)) & 0x33333333u;
    v = (v | (v << 1)) & 0x55555555u;
    return v;
}
RJ_HD uint32_t compact16(uint32_t v) {
    v &= 0x55555555u;
    v = (v | (v >> 1)) & 0x33333333u;
    v = (v | (v >> 2)) & 0x0F0F0F0Fu;
    v = (v | (v >> 4)) & 0x00FF00FFu;
    v = (v | (v >> 8)) & 0x0000FFFFu;
    return v;
}
RJ_HD uint32_t morton_key(uint32_t qx, uint32_t qy) {
    return spread16(qx >> kMortonShift) | (spread16(qy >> kMortonShift) << 1);
}
// Point cells: the lattice is cut into 2^L x 2^L cells numbered in Morton
// order; because the points are sorted by the Morton key, every cell of
// every level L <= 10 is a contiguous range of the sorted points.
RJ_HD uint32_t cell_of(uint32_t qx, uint32_t qy, int L) {
    return spread16(qx >> (kLatticeBits - L)) | (spread16(qy >> (kLatticeBits - L)) << 1);
}
RJ_HD uint32_t cell_x(uint32_t c) { return compact16(c); }
RJ_HD uint32_t cell_y(uint32_t c) { return compact16(c >> 1); }

// Pixel range [lo, hi] (inclusive) covered by cell column/row cc (level L)
// of a canvas side of n pixels: the pixels whose lattice extent meets the cell.
RJ_HD int64_t cell_pix_lo(int64_t cc, int64_t n, int L) { return pix(cc << (kLatticeBits - L), n); }
RJ_HD int64_t cell_pix_hi(int64_t cc, int64_t n, int L) { return pix(((cc + 1) << (kLatticeBits - L)) - 1, n); }

// S5 supercover (reading Z6, O9): pixel columns [i0, i1] of row r touched by
// edge (xa,ya)-(xb,yb): clip the segment to the row's closed lattice band
// y in [max(qlo(r), ymin), min(qhi(r), ymax)]; its real x-extent [xl, xr]
// meets pixel i's closed extent [qlo(i), qhi(i)] (integers) iff
// qlo(i) <= floor(xr) and qhi(i) >= ceil(xl), i.e. pix(ceil(xl)) <= i <=
// pix(floor(xr)).  That range is empty only when the clipped segment lies in
// the open gap (qhi(i), qlo(i+1)) between two pixels' extents; a nearly
// vertical edge whose x-extent falls strictly between two consecutive
// lattice values INSIDE one pixel's extent (ceil(xl) > floor(xr), same
// pixel) touches that pixel.  Coordinate 2^30 and beyond is excluded.
RJ_HD bool supercover_cols(int64_t xa, int64_t ya, int64_t xb, int64_t yb, int64_t r, int64_t W, int64_t H,
                           int64_t &i0, int64_t &i1) {
    const int64_t ymin = ya < yb ? ya : yb, ymax = ya < yb ? yb : ya;
    const int64_t ql = qlo(r, H), qh = qhi(r, H);
    const int64_t ylo = ql > ymin ? ql : ymin, yhi = qh < ymax ? qh : ymax;
    int64_t cl, fr;
    if (ya == yb) {
        cl = xa < xb ? xa : xb;
        fr = xa < xb ? xb : xa;
    } else {
        int64_t d = yb - ya, dx = xb - xa, base = xa * d;
        int64_t n1 = base + dx * (ylo - ya), n2 = base + dx * (yhi - ya);
        if (d < 0) { d = -d; n1 = -n1; n2 = -n2; }
        const int64_t c1 = ceil_div(n1, d), c2 = ceil_div(n2, d), f1 = floor_div(n1, d), f2 = floor_div(n2, d);
        cl = c1 < c2 ? c1 : c2;
        fr = f1 > f2 ? f1 : f2;
    }
    if (cl >= kOne) return false;
    if (fr > kOne - 1) fr = kOne - 1;
    i0 = pix(cl, W);
    i1 = pix(fr, W);
    return i0 <= i1;
}

// Rows of the supercover band of an edge / polygon with y-extent [ymin, ymax]:
// [pix(ymin), pix(min(ymax, 2^30 - 1))], none when ymin >= 2^30.
RJ_HD int64_t band_rows(int64_t ymin, int64_t ymax, int64_t H) {
    return ymin >= kOne ? 0 : pix(ymax < kOne - 1 ? ymax : kOne - 1, H) - pix(ymin, H) + 1;
}

}  // namespace rj

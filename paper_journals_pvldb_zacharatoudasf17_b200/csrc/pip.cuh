// pip.cuh -- exact even-odd point-in-polygon walk through the S6 edge grid
// (Proc. JoinPoint; grid index P:906-917), shared by the
// fused point pass (boundary points, index join) and the streamed query.
//
// Cell (gx, gy) of the 1024 x 1024 grid lists, per polygon P whose MBR meets
// it, every non-horizontal edge of P whose y-extent overlaps the cell's rows
// and that can toggle the half-open PNPOLY ray of a point in the cell
// (reading Z4) -- a rightward ray in the cells from the middle of P's MBR on,
// a leftward one left of it (reading Z25; bit 31 of the polygon id).
// Entries are sorted (flag, edge id), so they group by polygon; each entry is
// inlined as the upward-oriented edge (xl, yl, dx = xu - xl, yu), yl < yu,
// + polygon id.
#pragma once
#include "rj_geom.cuh"

namespace rj {

constexpr uint32_t kPipNone = 0xFFFFFFFFu;

// Returns the first containing polygon (kPipNone if none); every further
// containing polygon (overlapping polygons) is passed to extra(P).
template <class F>
__device__ __forceinline__ uint32_t grid_pip(const uint32_t *__restrict__ grid_off,
                                             const uint32_t *__restrict__ grid_poly,
                                             const int4 *__restrict__ grid_edge, uint32_t px, uint32_t py,
                                             F &&extra) {
    const uint32_t cell = (py >> kGridShift) * kGrid + (px >> kGridShift);
    const uint32_t b = __ldg(&grid_off[cell]), e = __ldg(&grid_off[cell + 1]);
    uint32_t cur = kPipNone, par = 0, first = kPipNone;
    const int X = (int)px, Y = (int)py;                    // lattice coordinates < 2^30
    for (uint32_t k = b; k < e; ++k) {
        const uint32_t PL = __ldg(&grid_poly[k]);
        const uint32_t P = PL & 0x7FFFFFFFu;
        const int4 E = __ldg(&grid_edge[k]);
        if (P != cur) {
            if (par) {
                if (first == kPipNone) first = cur;
                else extra(cur);
            }
            cur = P;
            par = 0;
        }
        // PNPOLY toggle (O3, half-open in y) of the edge oriented upwards:
        // yl <= py < yu and px < the crossing's x, i.e.
        // (px - xl)(yu - yl) < (xu - xl)(py - yl); every factor fits 31 bits
        // plus sign, so each product is one exact 32 x 32 -> 64-bit multiply
        // A leftward-ray entry (bit 31) toggles on the complement, X* <= px:
        // a closed ring has an even number of edges straddling the row, so
        // both rays give the same parity, ties included (reading Z25).
        if (E.y <= Y && Y < E.w) {
            const long long lhs = (long long)(X - E.x) * (E.w - E.y);
            const long long rhs = (long long)E.z * (Y - E.y);
            par ^= (lhs < rhs ? 1u : 0u) ^ (PL >> 31);
        }
    }
    if (par) {
        if (first == kPipNone) first = cur;
        else extra(cur);
    }
    return first;
}

}  // namespace rj

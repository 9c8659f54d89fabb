// pip.cuh -- exact even-odd point-in-polygon walk through the S6 edge grid
// (Proc. JoinPoint; grid index P:906-917), shared by the
// fused point pass (boundary points, index join) and the streamed query.
//
// Cell (gx, gy) of the 1024 x 1024 grid lists every non-horizontal edge whose
// y-extent overlaps the cell's rows and that lies (partly) at or right of the
// cell inside its polygon's MBR: exactly the edges that can toggle the
// half-open PNPOLY ray of a point in the cell (reading Z4).  Entries are
// sorted by edge id, so they group by polygon; each entry is inlined as
// (xa, ya, xb, yb) + polygon id.
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
    const int64_t X = px, Y = py;
    for (uint32_t k = b; k < e; ++k) {
        const uint32_t P = __ldg(&grid_poly[k]);
        const int4 E = __ldg(&grid_edge[k]);
        if (P != cur) {
            if (par) {
                if (first == kPipNone) first = cur;
                else extra(cur);
            }
            cur = P;
            par = 0;
        }
        // PNPOLY toggle (half-open in y), exact in int64
        if ((E.y > (int)py) != (E.w > (int)py)) {
            const int64_t lhs = (X - E.x) * (int64_t)(E.w - E.y);
            const int64_t rhs = (int64_t)(E.z - E.x) * (Y - E.y);
            if (E.w > E.y ? lhs < rhs : lhs > rhs) par ^= 1u;
        }
    }
    if (par) {
        if (first == kPipNone) first = cur;
        else extra(cur);
    }
    return first;
}

}  // namespace rj

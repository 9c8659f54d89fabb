// work.cu -- work-item planning of the fused point pass (host runtime).
//
// A query at canvas W x H uses point cells of level L (2^L x 2^L lattice
// cells) whose pixel footprint is ~16-32 pixels a side, so one warp's tile
// fits in shared memory.  Work items are contiguous ranges of the sorted
// points: a run of consecutive light cells (<= chunk points together), or
// one chunk of a heavy cell.  Items depend only on the loaded points and L,
// so they are planned once per level and cached.
#include <algorithm>

#include "rj_internal.cuh"

namespace rj {

int choose_level(int W, int H, int target) {
    // smallest L whose cells span <= target pixels a side (capped at level 10)
    const int side = std::max(W, H);
    int L = 0;
    while (L < kMaxLevel && (side + (1 << L) - 1) / (1 << L) > target) ++L;
    return L;
}

void drop_items(Ctx *c) {
    for (int L = 0; L <= kMaxLevel; ++L) {
        dfree(c, c->items[L]);
        dfree(c, c->cell_bits[L]);
        c->n_items[L] = 0;
        c->items_chunk[L] = 0;
    }
    c->h_cell_off.clear();
}

rj_status items_for_level(Ctx *c, int L) {
    if (c->items[L].p && c->items_chunk[L] == c->chunk) return RJ_OK;
    if (c->h_cell_off.empty()) {
        c->h_cell_off.resize((size_t)kCells10 + 1);
        RJ_CUDA(c, cudaMemcpyAsync(c->h_cell_off.data(), c->cell_off.p, ((size_t)kCells10 + 1) * 4,
                                   cudaMemcpyDeviceToHost, c->stream));
        RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    }
    const uint64_t ncell = 1ull << (2 * L);
    const int sh = 2 * (kMaxLevel - L);
    const uint64_t CH = (uint64_t)std::max<int64_t>(64, c->chunk);
    const uint32_t *off = c->h_cell_off.data();
    std::vector<int4> items;
    int64_t gb = -1, ge = -1;       // open group: cells [gb, ge)
    uint64_t gpts = 0, gcells = 0;
    // a group's cost is ~ its points plus a fixed tile setup/reduce per cell:
    // cap both so that no single item dominates the tail of the pass
    const uint64_t max_cells = 8;
    auto flush = [&]() {
        if (gb >= 0) items.push_back(make_int4((int)gb, (int)ge, (int)off[(uint64_t)gb << sh], (int)off[(uint64_t)ge << sh]));
        gb = -1;
        gpts = 0;
        gcells = 0;
    };
    for (uint64_t cc = 0; cc < ncell; ++cc) {
        const uint64_t b = off[cc << sh], e = off[(cc + 1) << sh], m = e - b;
        if (!m) continue;
        if (m > CH) {
            flush();
            const uint64_t k = (m + CH - 1) / CH;
            for (uint64_t j = 0; j < k; ++j)
                items.push_back(make_int4((int)cc, (int)cc + 1, (int)(b + m * j / k), (int)(b + m * (j + 1) / k)));
            continue;
        }
        if (gb >= 0 && (gpts + m > CH || (int64_t)cc - ge > 16 || gcells >= max_cells)) flush();
        if (gb < 0) gb = (int64_t)cc;
        ge = (int64_t)cc + 1;
        gpts += m;
        gcells += 1;
    }
    flush();
    // Guided tail: CTAs take items in order from one counter, so the last
    // items decide how unevenly the persistent grid finishes (a 64k-point
    // item is ~40 us of one CTA's stream).  The items holding the last ~one
    // item per CTA of points are re-cut into single cells and <= CH/8-point
    // chunks, so every CTA that finishes its last large item finds small
    // ones -- the points are the same, only the final items are finer.
    {
        uint64_t total = 0;
        for (const int4 &I : items) total += (uint64_t)(I.w - I.z);
        const uint64_t tail_pts = std::min<uint64_t>(total / 4, (uint64_t)c->num_sms * 2 * CH);
        const uint64_t cht = std::max<uint64_t>(2048, CH / 8);
        size_t k = items.size();
        uint64_t acc = 0;
        while (k > 0 && acc < tail_pts) {
            --k;
            acc += (uint64_t)(items[k].w - items[k].z);
        }
        std::vector<int4> tail;
        for (size_t i = k; i < items.size(); ++i) {
            const int4 I = items[i];
            for (int64_t cc = I.x; cc < I.y; ++cc) {
                const uint64_t b = std::max<uint64_t>((uint64_t)I.z, off[(uint64_t)cc << sh]);
                const uint64_t e = std::min<uint64_t>((uint64_t)I.w, off[(uint64_t)(cc + 1) << sh]);
                if (b >= e) continue;
                const uint64_t m = e - b, parts = (m + cht - 1) / cht;
                for (uint64_t j = 0; j < parts; ++j)
                    tail.push_back(make_int4((int)cc, (int)cc + 1, (int)(b + m * j / parts), (int)(b + m * (j + 1) / parts)));
            }
        }
        items.resize(k);
        items.insert(items.end(), tail.begin(), tail.end());
    }
    // non-empty point cells of the level as a bitmask (the polygon pass skips
    // span pieces of empty cells with one L1-friendly word load)
    std::vector<uint32_t> bits((ncell + 31) / 32, 0u);
    for (uint64_t cc = 0; cc < ncell; ++cc)
        if (off[(cc + 1) << sh] != off[cc << sh]) bits[cc >> 5] |= 1u << (cc & 31);
    dfree(c, c->cell_bits[L]);
    if (dalloc(c, c->cell_bits[L], bits.size() * 4)) return set_error(c, RJ_ERR_OOM, "cell mask allocation failed");
    RJ_CUDA(c, cudaMemcpyAsync(c->cell_bits[L].p, bits.data(), bits.size() * 4, cudaMemcpyHostToDevice, c->stream));
    dfree(c, c->items[L]);
    if (dalloc(c, c->items[L], std::max<size_t>(1, items.size()) * sizeof(int4)))
        return set_error(c, RJ_ERR_OOM, "work item allocation failed");
    if (!items.empty())
        RJ_CUDA(c, cudaMemcpyAsync(c->items[L].p, items.data(), items.size() * sizeof(int4), cudaMemcpyHostToDevice,
                                   c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    c->n_items[L] = (uint32_t)items.size();
    c->items_chunk[L] = c->chunk;
    return RJ_OK;
}

}  // namespace rj

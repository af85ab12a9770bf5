// bottomup.cuh — the bottom-up BFS step over the in-CGR with early exit (north_star's direction optimisation;
// SURVEY §8 a9; not in the paper).  For every unvisited vertex v, v's IN-record is decoded until the first
// in-neighbour in the frontier F: intervals are tested as frontier-bitmap word ranges (32 parents per test), residuals
// as single bits, four probes in flight per batch; decoding stops at the first hit.
//
// A warp owns one 32-vertex word at a time (grid-stride), lane = vertex id, so the found mask is written to N with
// one plain store (no atomics).  In-records are read from global memory through the read-only path: most scans stop
// after a few codewords, so staging whole records through shared memory (measured) only adds copy work.
#pragma once
#include "apps.cuh"
#include "expand.cuh"

namespace gcgt_dev {

__device__ __forceinline__ bool frontier_range(const uint32_t* __restrict__ F, uint32_t s, uint32_t len) {
    const uint32_t e = s + len;
    while (s < e) {
        const uint32_t b0 = s & 31, nb = min(32u - b0, e - s);
        if (__ldg(F + (s >> 5)) & ((nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0)) return true;
        s += nb;
    }
    return false;
}

// Residual scan: cnt residuals, the first anchored at v, four frontier probes in flight per batch; stops at the
// first hit (or when *stop becomes non-zero).  got += residuals decoded.
template <int K>
__device__ __forceinline__ bool bu_residuals(GBitReader& r, uint32_t v, uint32_t cnt, const uint32_t* __restrict__ F,
                                             uint32_t& got, const volatile uint32_t* stop = nullptr) {
    if (cnt == 0) return false;
    uint32_t cur = unmap_first32(v, r.template next<K>());
    bool found = (__ldg(F + (cur >> 5)) >> (cur & 31)) & 1u;
    uint32_t i = 1;
    // whole batches of four: four decodes, then four frontier probes in flight together, one exit test
    for (; !found && i + 4 <= cnt; i += 4) {
        if (stop && *stop) break;
        uint32_t id[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            cur += (uint32_t)r.template next<K>();
            id[k] = cur;
        }
        uint32_t fw[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) fw[k] = __ldg(F + (id[k] >> 5));
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) found |= ((fw[k] >> (id[k] & 31)) & 1u) != 0;
    }
    for (; !found && i < cnt; i++) {  // tail
        cur += (uint32_t)r.template next<K>();
        found = (__ldg(F + (cur >> 5)) >> (cur & 31)) & 1u;
    }
    got += i;
    return found;
}

// Deferred bottom-up hubs: a vertex whose in-record has more than hub_segs residual segments (and no frontier parent
// in its interval area) is queued; its segments are then scanned by the whole grid (bu_hub_kernel), one per lane,
// with a per-vertex "found" flag that stops the other lanes' scans — the bottom-up analogue of the top-down hub pass.
struct BuHubs {
    HubEntry* q;
    unsigned long long* ctr;  // (entries << 32) | segments
    uint32_t* done;           // per entry: a frontier parent was found
    uint32_t hub_segs;
};

// In-record scan of v from reader r: true at the first in-neighbour in F.  na / nb: arcs decoded / bits consumed.
template <int K, bool SEG>
__device__ __forceinline__ bool bu_scan(GBitReader& r, uint64_t p0, uint64_t p1, uint32_t v, uint32_t min_len,
                                        uint32_t seg_bits, const uint32_t* __restrict__ F, const BuHubs& hubs,
                                        uint32_t& na, uint32_t& nb) {
    uint32_t deg = 0, got = 0;
    if (!SEG) deg = (uint32_t)(r.template next<K>() - 1);
    const uint32_t itv = (uint32_t)(r.template next<K>() - 1);
    uint32_t prev_end = 0;
    bool found = false;
    for (uint32_t i = 0; i < itv && !found; i++) {
        const uint64_t g = r.template next<K>();
        const uint32_t len = (uint32_t)(r.template next<K>() - 1) + min_len;
        const uint32_t start = i == 0 ? unmap_first32(v, g) : prev_end + (uint32_t)g;
        found = frontier_range(F, start, len);
        prev_end = start + len - 1;
        got += len;
    }
    uint64_t pend;
    if (found) {
        pend = r.pos();
    } else if (!SEG) {
        found = bu_residuals<K>(r, v, (uint32_t)(deg - got), F, got);
        pend = r.pos();
    } else {
        const uint32_t nseg = (uint32_t)(r.template next<K>() - 1);
        const uint64_t base = r.pos();
        pend = base;
        if (hubs.q && nseg > hubs.hub_segs) {  // long in-record: its segments go to the grid-wide pass
            const unsigned long long old = atomicAdd(hubs.ctr, (1ull << 32) | (unsigned long long)nseg);
            hubs.q[old >> 32] = HubEntry{base, p1, v, (uint32_t)(old & 0xffffffffu), nseg, 0};
            hubs.done[old >> 32] = 0;
            na += got;
            nb += (uint32_t)(pend - p0);
            return false;
        }
        for (uint32_t sg = 0; sg < nseg && !found; sg++) {
            r.init(r.src, r.j0, base + (uint64_t)sg * seg_bits);
            found = bu_residuals<K>(r, v, (uint32_t)(r.template next<K>() - 1), F, got);
            pend = r.pos();
        }
    }
    na += got;
    nb += (uint32_t)(pend - p0);
    return found;
}

template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock, 6) bu_kernel(const uint64_t* __restrict__ W, Offs offs, uint32_t min_len,
                                                       uint32_t seg_bits, const uint32_t* __restrict__ V,
                                                       const uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                                                       uint64_t lo, uint64_t hi, const uint32_t* __restrict__ dir,
                                                       unsigned long long* st, BuHubs hubs) {
    if (*dir != 1) return;
    const uint32_t lane = lane_id();
    uint32_t nv = 0, na = 0, nb = 0;
    const uint64_t w_lo = lo >> 5, w_hi = (hi + 31) >> 5;
    for (uint64_t w = w_lo + (((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5); w < w_hi;
         w += ((uint64_t)gridDim.x * blockDim.x) >> 5) {
        const uint64_t v0 = w * 32;
        uint32_t unv = ~__ldg(V + w);
        if (v0 < lo) unv &= 0xffffffffu << (lo - v0);
        if (hi - v0 < 32) unv &= (1u << (hi - v0)) - 1;
        if (!unv) continue;
        const bool act = (unv >> lane) & 1u;
        const uint32_t v = (uint32_t)(v0 + lane);
        uint64_t p0 = 0, p1 = 0;
        if (act) {
            p0 = offs(v);
            p1 = offs(v + 1);
        }
        bool found = false;
        if (act) {
            nv++;
            GBitReader r;
            r.init(reinterpret_cast<const uint32_t*>(W), 0, p0);
            found = bu_scan<K, SEG>(r, p0, p1, v, min_len, seg_bits, F, hubs, na, nb);
        }
        const uint32_t fb = __ballot_sync(0xffffffffu, found);
        if (lane == 0 && fb) N[w] = fb;
        __syncwarp();
    }
    add_stats3(st, nv, na, nb);
}

// The level's deferred bottom-up hubs: flattened segments over the whole grid, one per lane (read from global memory:
// most scans stop after a few probes).  The first lane to find a frontier parent sets the entry's flag and the
// vertex's bit in N; lanes check the flag before and during their segment.
template <int K>
__global__ void __launch_bounds__(kBlock) bu_hub_kernel(const uint64_t* __restrict__ W, uint32_t seg_bits,
                                                        const uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                                                        const uint32_t* __restrict__ dir, BuHubs hubs,
                                                        unsigned long long* st) {
    if (*dir != 1) return;
    const unsigned long long hc = *(volatile unsigned long long*)hubs.ctr;
    if (hc == 0) return;
    const uint32_t lane = lane_id();
    const uint32_t nh = (uint32_t)(hc >> 32), S = (uint32_t)(hc & 0xffffffffu);
    uint32_t na = 0;
    const uint64_t gw0 = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) & ~31ull;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t jb = gw0; jb < S; jb += stride) {
        const uint32_t j = (uint32_t)jb + lane;
        const uint32_t k = warp_find_hub(hubs.q, nh, (uint32_t)jb, min(j, S - 1));
        if (j >= S) continue;
        const HubEntry e = hubs.q[k];
        volatile uint32_t* flag = hubs.done + k;
        if (*flag) continue;
        GBitReader r;
        r.init(reinterpret_cast<const uint32_t*>(W), 0, e.base + (uint64_t)(j - e.seg_off) * seg_bits);
        uint32_t got = 0;
        const bool found = bu_residuals<K>(r, e.u, (uint32_t)(r.template next<K>() - 1), F, got, flag);
        na += got;
        if (found && atomicExch(hubs.done + k, 1u) == 0) red_or(N + (e.u >> 5), 1u << (e.u & 31));
    }
    add_stats3(st, 0, na, 0);
}

}  // namespace gcgt_dev

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

// ---- flat bottom-up: lane per 32-vertex word, flat scan loop -------------------------------------------------------
// bu_kernel gives each lane one vertex of the warp's 32-vertex word and the warp waits for its longest scan (early exits
// differ by orders of magnitude).  Here a lane owns a whole word and scans its unvisited vertices one after another in
// ONE flat loop: per iteration every busy lane takes one step of its current in-record -- the header, up to two
// intervals (range tests on F), the segment count, a segment's count, or up to four residuals (four probes in flight)
// -- and a lane whose vertex is finished moves to the next unvisited vertex of its word at once: consecutive vertices
// have consecutive records, so the next record is usually already in L1.  A lane whose word is finished writes the
// word's found mask to N (one plain store) and takes the next word of the warp's chunk.  The codewords of a step are
// decoded by the same unrolled code for every phase, so only the short interpretation diverges.
enum : uint32_t { kIdle = 0, kOpen, kHdr, kItv, kNseg, kSegStart, kRes };

template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock, 4) bu_flat_kernel(const uint64_t* __restrict__ W, Offs offs, uint32_t min_len,
                                                            uint32_t seg_bits, const uint32_t* __restrict__ V,
                                                            const uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                                                            uint64_t lo, uint64_t hi, const uint32_t* __restrict__ dir,
                                                            unsigned long long* st, BuHubs hubs) {
    if (*dir != 1) return;
    const uint32_t lane = lane_id();
    const uint32_t* W32 = reinterpret_cast<const uint32_t*>(W);
    uint32_t nv = 0, na = 0, nb = 0;
    const uint64_t w_lo = lo >> 5, w_hi = (hi + 31) >> 5;
    const uint64_t nwarp = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    uint64_t chunk = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;  // 32-word chunks, grid-stride
    uint64_t wbase = 0;
    uint32_t myunv = 0, wmask = 0;  // lane l: unvisited vertices of chunk word wbase + l; chunk words not yet taken
    bool more = true;
    // lane state: the word being scanned (w, its remaining unvisited bits m, found bits fm), the vertex, the reader
    GBitReader r;
    uint64_t w = 0;
    uint32_t m = 0, fm = 0;
    uint32_t ph = kIdle, v = 0, rem = 0, cur = 0, seg = 0, nseg = 0, deg = 0, got = 0;
    bool first = false;
    uint64_t p0 = 0, sbase = 0;
    for (;;) {
        // ---- idle lanes take the next words with unvisited vertices (warp-uniform control flow)
        uint32_t need = __ballot_sync(0xffffffffu, ph == kIdle);
        while (need && (wmask || more)) {
            if (!wmask) {
                const uint64_t wb = w_lo + chunk * 32;
                chunk += nwarp;
                if (wb >= w_hi) {
                    more = false;
                    break;
                }
                wbase = wb;
                const uint64_t ww = wb + lane;
                myunv = 0;
                if (ww < w_hi) {
                    const uint64_t v0 = ww * 32;
                    myunv = ~__ldg(V + ww);
                    if (v0 < lo) myunv &= 0xffffffffu << (lo - v0);
                    if (hi - v0 < 32) myunv &= (1u << (hi - v0)) - 1;
                }
                wmask = __ballot_sync(0xffffffffu, myunv != 0);
                continue;
            }
            const uint32_t nn = __popc(need), np = __popc(wmask), tk = min(nn, np);
            uint32_t src_lane = 0;
            const bool me = (need >> lane) & 1u;
            const uint32_t j = __popc(need & lanemask_lt());
            if (me && j < tk) src_lane = __fns(wmask, 0, (int)j + 1);
            const uint32_t mm = __shfl_sync(0xffffffffu, myunv, src_lane);
            if (me && j < tk) {
                w = wbase + src_lane;
                m = mm;
                fm = 0;
                ph = kOpen;
            }
            wmask = tk == np ? 0u : wmask & (0xffffffffu << __fns(wmask, 0, (int)tk + 1));
            need = tk == nn ? 0u : need & (0xffffffffu << __fns(need, 0, (int)tk + 1));
        }
        if (!__any_sync(0xffffffffu, ph != kIdle)) break;
        // ---- open the next unvisited vertex of the lane's word
        if (ph == kOpen) {
            const uint32_t b = __ffs(m) - 1;
            m &= m - 1;
            v = (uint32_t)(w * 32 + b);
            p0 = offs(v);
            const uint64_t p1 = offs(v + 1);
            nv++;
            got = 0;
            if (p0 == p1) ph = kOpen;  // no in-arcs: not found; the word's next vertex (or the word is done)
            else {
                r.init(W32, 0, p0);
                ph = kHdr;
            }
            if (ph == kOpen && !m) {
                if (fm) N[w] = fm;
                ph = kIdle;
            }
        }
        // ---- per-lane step
        if (ph == kSegStart) r.init(W32, 0, sbase + (uint64_t)seg * seg_bits);
        uint32_t ncw = 0;
        if (ph == kHdr || ph == kNseg || ph == kSegStart) ncw = (ph == kHdr && !SEG) ? 2 : 1;
        else if (ph == kItv) ncw = rem >= 2 ? 4 : 2;
        else if (ph == kRes) ncw = min(rem, 4u);
        uint32_t x[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            x[k] = 0;
            if (k < ncw) {
                const uint64_t c = r.template next<K>();
                x[k] = (k == 0 && first) ? unmap_first32(v, c) : (uint32_t)c;
            }
        }
        bool found = false, done = false;
        if (ph == kRes) {
            uint32_t id[4];
#pragma unroll
            for (uint32_t k = 0; k < 4; k++) {
                cur = (k == 0 && first) ? x[0] : cur + x[k];
                id[k] = cur;
            }
            uint32_t fw[4];
#pragma unroll
            for (uint32_t k = 0; k < 4; k++) fw[k] = k < ncw ? __ldg(F + (id[k] >> 5)) : 0u;
#pragma unroll
            for (uint32_t k = 0; k < 4; k++) found |= ((fw[k] >> (id[k] & 31)) & 1u) != 0;
            first = false;
            rem -= ncw;
            got += ncw;
            if (rem == 0) {
                if (!SEG) done = true;
                else if (++seg == nseg) done = true;
                else ph = kSegStart;
            }
        } else if (ph == kItv) {
#pragma unroll
            for (uint32_t k = 0; k < 4; k += 2) {
                if (k < ncw) {
                    const uint32_t start = (k == 0 && first) ? x[0] : cur + x[k];
                    const uint32_t len = x[k + 1] - 1 + min_len;
                    found |= frontier_range(F, start, len);
                    cur = start + len - 1;
                    got += len;
                }
            }
            first = false;
            rem -= ncw >> 1;
            if (rem == 0) {
                if (SEG) ph = kNseg;
                else if (deg > got) { ph = kRes; rem = deg - got; first = true; }
                else done = true;
            }
        } else if (ph == kHdr) {
            uint32_t itv;
            if (SEG) itv = x[0] - 1;
            else { deg = x[0] - 1; itv = x[1] - 1; }
            if (itv) { ph = kItv; rem = itv; first = true; }
            else if (SEG) ph = kNseg;
            else if (deg) { ph = kRes; rem = deg; first = true; }
            else done = true;
        } else if (ph == kNseg) {
            nseg = x[0] - 1;
            sbase = r.pos();
            seg = 0;
            if (nseg == 0) done = true;
            else if (hubs.q && nseg > hubs.hub_segs) {  // long in-record: its segments go to the grid-wide pass
                const unsigned long long old = atomicAdd(hubs.ctr, (1ull << 32) | (unsigned long long)nseg);
                hubs.q[old >> 32] = HubEntry{sbase, offs(v + 1), v, (uint32_t)(old & 0xffffffffu), nseg, 0};
                hubs.done[old >> 32] = 0;
                done = true;
            } else ph = kSegStart;
        } else if (ph == kSegStart) {
            rem = x[0] - 1;
            first = true;
            ph = rem ? kRes : kIdle;  // (R19: a segment holds at least one residual)
            if (!rem) done = true;
        }
        if (found || done) {
            if (found) fm |= 1u << (v & 31);
            na += got;
            nb += (uint32_t)(r.pos() - p0);
            rem = 0;
            first = false;
            ph = kOpen;
            if (!m) {  // the lane's word is finished
                if (fm) N[w] = fm;
                ph = kIdle;
            }
        }
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

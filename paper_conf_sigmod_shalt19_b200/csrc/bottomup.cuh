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

// In-record scan of v from reader r: true at the first in-neighbour in F.  na / nb: arcs decoded / bits consumed.
template <int K, bool SEG>
__device__ __forceinline__ bool bu_scan(GBitReader& r, uint64_t p0, uint64_t p1, uint32_t v, uint32_t min_len,
                                        uint32_t seg_bits, const uint32_t* __restrict__ F, uint32_t& na,
                                        uint32_t& nb) {
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
                                                       unsigned long long* st) {
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
            found = bu_scan<K, SEG>(r, p0, p1, v, min_len, seg_bits, F, na, nb);
        }
        const uint32_t fb = __ballot_sync(0xffffffffu, found);
        if (lane == 0 && fb) N[w] = fb;
        __syncwarp();
    }
    add_stats3(st, nv, na, nb);
}

}  // namespace gcgt_dev

#pragma once
#include "apps.cuh"
#include "expand.cuh"

namespace gcgt_dev {

// csr_bfs.cuh — uncompressed-CSR BFS on the same B200 (§8 f3).
//
// The paper compares GCGT with an uncompressed GPU BFS ("GPUCSR", Merrill et al.) and reports the
// decoding overhead (+54 % at 18.1x compression, Fig. 8 :1571-1578).  This is that baseline on B200, built from the
// same parts as the CGR path so that the ratio isolates decoding: the same frontier (bitmap F + queue of frontier
// words), the same filter (BfsApp: read-only visited pre-test, fire-and-forget atomicOr on N), the same contraction
// (commit_kernel) and direction choice (decide_body).  Only the expansion differs: neighbour ids are read from col[]:
//  * top-down: a warp takes batches of frontier words, lists their vertices, and flattens the arcs of 32 vertices at
//    a time over its lanes (coalesced col[] reads, four ids in flight per lane); vertices with more than
//    kCsrHub arcs go to a per-level hub queue whose kCsrChunk-arc chunks are spread over the whole grid;
//  * bottom-up: warp per 32-vertex word, lane per unvisited vertex scanning its in-list (the transpose, or col[]
//    itself on symmetric graphs) until the first frontier parent.

constexpr uint32_t kCsrHub = 4096;
constexpr uint32_t kCsrChunk = 1024;

struct CsrHubEntry {
    uint64_t beg;        // first arc
    uint32_t deg;
    uint32_t chunk_off;  // first flattened chunk index (entries are ordered by chunk_off)
};

struct CsrSmem {
    uint32_t w[32], b[32], pre[33], dpre[33];
    uint64_t beg[32];
};

template <class Front>
__global__ void __launch_bounds__(kBlock, 4) csr_expand_kernel(const uint64_t* __restrict__ row,
                                                               const uint32_t* __restrict__ col, Front fr, BfsApp app,
                                                               unsigned long long* cursor, CsrHubEntry* hubq,
                                                               unsigned long long* hub_ctr, const uint32_t* dir,
                                                               unsigned long long* st) {
    __shared__ CsrSmem smem[kWarps];
    const uint32_t wid = threadIdx.x >> 5, lane = lane_id();
    CsrSmem& sm = smem[wid];
    uint64_t nv = 0, na = 0;
    if (!(dir && *dir)) {
        const uint64_t qlen = fr.size();
        uint64_t wpb = qlen / ((uint64_t)gridDim.x * kWarps * 4);
        wpb = wpb < 1 ? 1 : (wpb > 8 ? 8 : wpb);
        unsigned long long next = 0;
        if (lane == 0) next = atomicAdd(cursor, (unsigned long long)wpb);
        for (;;) {
            const uint64_t base = __shfl_sync(0xffffffffu, next, 0);
            if (base >= qlen) break;
            if (lane == 0) next = atomicAdd(cursor, (unsigned long long)wpb);
            uint32_t w = 0, bits = 0;
            if (lane < wpb && base + lane < qlen) fr.get(base + lane, w, bits);
            uint32_t incl = __popc(bits);
            for (int o = 1; o < 32; o <<= 1) {
                const uint32_t t = __shfl_up_sync(0xffffffffu, incl, o);
                if (lane >= (uint32_t)o) incl += t;
            }
            sm.w[lane] = w;
            sm.b[lane] = bits;
            sm.pre[lane + 1] = incl;
            if (lane == 0) sm.pre[0] = 0;
            __syncwarp();
            const uint32_t total = sm.pre[32];
            for (uint32_t t0 = 0; t0 < total; t0 += 32) {
                const uint32_t j = t0 + lane;
                uint64_t beg = 0;
                uint32_t deg = 0;
                if (j < total) {
                    uint32_t lo = 0, hi = 31;  // owner word: largest o with pre[o] <= j
                    while (lo < hi) {
                        const uint32_t mid = (lo + hi + 1) >> 1;
                        if (sm.pre[mid] <= j) lo = mid; else hi = mid - 1;
                    }
                    const uint32_t u = sm.w[lo] * 32 + __fns(sm.b[lo], 0, (int)(j - sm.pre[lo]) + 1);
                    beg = ldg64(row + u);
                    const uint64_t d = ldg64(row + u + 1) - beg;
                    nv++;
                    if (d > kCsrHub) {  // hub: its arcs go to the whole grid
                        const uint32_t nch = (uint32_t)((d + kCsrChunk - 1) / kCsrChunk);
                        const unsigned long long old = atomicAdd(hub_ctr, (1ull << 32) | (unsigned long long)nch);
                        hubq[old >> 32] = CsrHubEntry{beg, (uint32_t)d, (uint32_t)(old & 0xffffffffu)};
                    } else {
                        deg = (uint32_t)d;
                    }
                }
                uint32_t dincl = deg;
                for (int o = 1; o < 32; o <<= 1) {
                    const uint32_t t = __shfl_up_sync(0xffffffffu, dincl, o);
                    if (lane >= (uint32_t)o) dincl += t;
                }
                sm.beg[lane] = beg;
                sm.dpre[lane + 1] = dincl;
                if (lane == 0) sm.dpre[0] = 0;
                __syncwarp();
                const uint32_t A = sm.dpre[32];
                na += lane == 0 ? A : 0;
                uint32_t o = 0;  // owner of the lane's current arc (arcs only move forward)
                for (uint32_t k0 = 0; k0 < A; k0 += 128) {
                    uint32_t v[4];
                    uint32_t nb = 0;
#pragma unroll
                    for (uint32_t r = 0; r < 4; r++) {
                        const uint32_t k = k0 + r * 32 + lane;
                        if (k < A) {
                            while (sm.dpre[o + 1] <= k) o++;
                            v[r] = __ldg(col + sm.beg[o] + (k - sm.dpre[o]));
                            nb = r + 1;
                        }
                    }
                    app.many(v, nb);
                }
                __syncwarp();
            }
            __syncwarp();
        }
    }
    add_stats3(st, nv, na, na * 32);  // the work cursor is reset by the contraction
}

// Hub arcs of the level: warp per kCsrChunk-arc chunk (grid-stride), lanes stride the chunk (coalesced).
__global__ void __launch_bounds__(kBlock) csr_hub_kernel(const uint32_t* __restrict__ col, const CsrHubEntry* hubq,
                                                         const unsigned long long* hub_ctr, BfsApp app, unsigned long long* st) {
    const uint32_t lane = lane_id();
    const unsigned long long hc = *(volatile const unsigned long long*)hub_ctr;
    const uint32_t nh = (uint32_t)(hc >> 32), S = (uint32_t)(hc & 0xffffffffu);
    uint64_t na = 0;
    for (uint64_t j = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5; j < S;
         j += ((uint64_t)gridDim.x * blockDim.x) >> 5) {
        uint32_t lo = 0, hi = nh - 1;  // entry: largest e with chunk_off <= j
        while (lo < hi) {
            const uint32_t mid = (lo + hi + 1) >> 1;
            if (hubq[mid].chunk_off <= j) lo = mid; else hi = mid - 1;
        }
        const CsrHubEntry e = hubq[lo];
        const uint64_t a0 = (uint64_t)(j - e.chunk_off) * kCsrChunk;
        const uint64_t rem = e.deg - a0;
        const uint32_t cnt = rem < kCsrChunk ? (uint32_t)rem : kCsrChunk;
        if (lane == 0) na += cnt;
        for (uint32_t k0 = 0; k0 < cnt; k0 += 128) {
            uint32_t v[4];
            uint32_t nb = 0;
#pragma unroll
            for (uint32_t r = 0; r < 4; r++) {
                const uint32_t k = k0 + r * 32 + lane;
                if (k < cnt) {
                    v[r] = __ldg(col + e.beg + a0 + k);
                    nb = r + 1;
                }
            }
            app.many(v, nb);
        }
    }
    add_stats3(st, 0, na, na * 32);
}

// Bottom-up level over the in-lists: warp per word, lane per unvisited vertex, stop at the first frontier parent.
__global__ void __launch_bounds__(kBlock) csr_bu_kernel(const uint64_t* __restrict__ row,
                                                        const uint32_t* __restrict__ col,
                                                        const uint32_t* __restrict__ V,
                                                        const uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                                                        uint64_t n, const uint32_t* __restrict__ dir, unsigned long long* st) {
    if (*dir != 1) return;
    const uint32_t lane = lane_id();
    const uint64_t nwv = (n + 31) >> 5;
    uint64_t nv = 0, na = 0;
    for (uint64_t w = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5; w < nwv;
         w += ((uint64_t)gridDim.x * blockDim.x) >> 5) {
        const uint64_t v0 = w * 32;
        uint32_t unv = ~__ldg(V + w);
        if (n - v0 < 32) unv &= (1u << (n - v0)) - 1;
        if (!unv) continue;
        bool found = false;
        if ((unv >> lane) & 1u) {
            const uint64_t v = v0 + lane;
            const uint64_t b = ldg64(row + v), e = ldg64(row + v + 1);
            nv++;
            uint64_t i = b;
            for (; i < e; i++) {
                const uint32_t u = __ldg(col + i);
                if ((__ldg(F + (u >> 5)) >> (u & 31)) & 1u) {
                    found = true;
                    i++;
                    break;
                }
            }
            na += i - b;
        }
        const uint32_t fb = __ballot_sync(0xffffffffu, found);
        if (lane == 0 && fb) N[w] = fb;
    }
    add_stats3(st, nv, na, na * 32);
}

}  // namespace gcgt_dev

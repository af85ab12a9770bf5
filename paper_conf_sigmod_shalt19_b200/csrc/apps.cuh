// apps.cuh — the filters of the traversal applications (Fig. 7).  The expansion engine hands
// every decoded neighbour (or interval run) of a frontier vertex u to the application between begin(u) and end():
//   range(s, len)  an interval run [s, s+len) (Alg. 2 l.23-32: expanded by word-granular operations here)
//   one(v)         one residual neighbour
//   many(v[4], n)  up to four residual neighbours whose probes can be in flight together
#pragma once
#include <cooperative_groups.h>
#include <cooperative_groups/reduce.h>

#include "device.cuh"

namespace gcgt_dev {
namespace cg = cooperative_groups;

// Applies fn(word, mask) to the 32-id words of the run [s, s+len).
template <class Fn>
__device__ __forceinline__ void for_words(uint32_t s, uint32_t len, Fn&& fn) {
    const uint32_t e = s + len;
    while (s < e) {
        const uint32_t b0 = s & 31, nb = min(32u - b0, e - s);
        fn(s >> 5, (nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0);
        s += nb;
    }
}

// BFS (Fig. 7(b)).  V (visited, levels <= d) is immutable during a level, so it is read through the read-only
// path; a new vertex is claimed by a fire-and-forget OR into the next-frontier bitmap N (REDG); levels are written by
// the contraction.  An interval is claimed 32 ids per reduction.
struct BfsApp {
    const uint32_t* __restrict__ V;
    uint32_t* __restrict__ N;
    uint32_t nfilter;  // 1: also skip targets an (L1-cached, possibly stale) read of N shows as already claimed
    // N only gains bits during a level, so a stale read can only under-report claims: filtering on it never drops
    // a discovery; it saves same-address reductions on popular targets (social graphs)
    __device__ __forceinline__ static uint32_t ld_n(const uint32_t* p) {
        uint32_t x;
        asm volatile("ld.global.ca.u32 %0, [%1];" : "=r"(x) : "l"(p));
        return x;
    }
    __device__ __forceinline__ void begin(uint32_t) {}
    __device__ __forceinline__ void end() {}
    __device__ __forceinline__ void vertex(uint32_t) {}
    __device__ __forceinline__ void claim(uint32_t w, uint32_t mask) {
        uint32_t cand = mask & ~__ldg(V + w);
        if (cand && nfilter) cand &= ~ld_n(N + w);
        if (cand) red_or(N + w, cand);
    }
    __device__ __forceinline__ void one(uint32_t v) { claim(v >> 5, 1u << (v & 31)); }
    __device__ __forceinline__ void many(const uint32_t (&v)[4], uint32_t n) {
        uint32_t m[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) m[k] = k < n ? __ldg(V + (v[k] >> 5)) : 0xffffffffu;
        if (nfilter) {
#pragma unroll
            for (uint32_t k = 0; k < 4; k++)
                if (!((m[k] >> (v[k] & 31)) & 1u)) m[k] |= ld_n(N + (v[k] >> 5));
        }
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            const uint32_t bit = 1u << (v[k] & 31);
            if (!(m[k] & bit)) red_or(N + (v[k] >> 5), bit);
        }
    }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for_words(s, len, [&](uint32_t w, uint32_t mask) { claim(w, mask); });
    }
};

#define GCGT_MANY_BY_ONE                                                         \
    __device__ __forceinline__ void many(const uint32_t (&v)[4], uint32_t n) {  \
        for (uint32_t k = 0; k < n; k++) one(v[k]);                              \
    }

// BC forward (Fig. 7(d), Brandes [9]): an arc u->v with v not in V (levels <= d) has level(v) = d+1, so
// sigma(v) += sigma(u); N collects level d+1.
struct BcFwdApp {
    const uint32_t* __restrict__ V;
    uint32_t* __restrict__ N;
    double* __restrict__ sigma;
    double su;
    __device__ __forceinline__ void begin(uint32_t u) { su = sigma[u]; }
    __device__ __forceinline__ void end() {}
    __device__ __forceinline__ void vertex(uint32_t) {}
    __device__ __forceinline__ void claim(uint32_t w, uint32_t mask) {
        const uint32_t cand = mask & ~__ldg(V + w);
        if (!cand) return;
        red_or(N + w, cand);
        for (uint32_t cb = cand; cb; cb &= cb - 1) atomicAdd(sigma + (uint64_t)w * 32 + (__ffs(cb) - 1), su);
    }
    __device__ __forceinline__ void one(uint32_t v) { claim(v >> 5, 1u << (v & 31)); }
    GCGT_MANY_BY_ONE
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for_words(s, len, [&](uint32_t w, uint32_t mask) { claim(w, mask); });
    }
};

// BC backward: delta(u) = sum_{w in out(u), d(w) = d(u)+1} sigma(u)/sigma(w) (1 + delta(w))  (Fig. 7(d)), computed as
// sigma(u) * sum X(w) with X(w) = (1 + delta(w)) / sigma(w) precomputed for the level d+1 vertices (bc_level_x): one
// random fp64 read per successor arc instead of two and a division.  Successors are tested on a bitmap of level d+1
// (n/8 bytes, L2-resident) instead of the 4n-byte levels array, four arcs' reads in flight together.  A vertex's arcs
// are split over tasks (interval area + segments), so each task adds its partial sum to delta(u) and bc(u)
// (u != source); delta is zeroed per source.  Zero partials are skipped, so exact zeros stay exact.
struct BcBwdApp {
    const uint32_t* __restrict__ LB;  // level d+1 bitmap
    const double* __restrict__ X;     // (1 + delta) / sigma of the level d+1 vertices
    const double* __restrict__ sigma;
    double* __restrict__ delta;
    double* __restrict__ bc;
    uint32_t source;
    uint32_t u;
    double acc;
    __device__ __forceinline__ void begin(uint32_t uu) {
        u = uu;
        acc = 0.0;
    }
    __device__ __forceinline__ void vertex(uint32_t) {}
    __device__ __forceinline__ void one(uint32_t w) {
        if ((__ldg(LB + (w >> 5)) >> (w & 31)) & 1u) acc += X[w];
    }
    __device__ __forceinline__ void many(const uint32_t (&v)[4], uint32_t n) {
        uint32_t m[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) m[k] = k < n ? __ldg(LB + (v[k] >> 5)) : 0u;
        double x[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) x[k] = ((m[k] >> (v[k] & 31)) & 1u) ? X[v[k]] : 0.0;
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) acc += x[k];
    }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for_words(s, len, [&](uint32_t w, uint32_t mask) {
            for (uint32_t b = __ldg(LB + w) & mask; b; b &= b - 1) acc += X[w * 32 + (__ffs(b) - 1)];
        });
    }
    __device__ __forceinline__ void end() {
        // lanes finishing tasks of the same vertex (a hub's segments sit side by side in the hub queue) first sum
        // their partials, so a vertex with 10^5 segments does not serialise 10^5 fp64 atomics on one address
        cg::coalesced_group act = cg::coalesced_threads();
        cg::coalesced_group same = cg::labeled_partition(act, u);
        const double sum = cg::reduce(same, acc, cg::plus<double>());
        if (same.thread_rank() == 0 && sum != 0.0) {
            const double d = sigma[u] * sum;
            atomicAdd(delta + u, d);
            if (u != source) atomicAdd(bc + u, d);
        }
    }
};

// ---- CC -------------------------------------------------------------------------------------------------------------
// Hooking (Fig. 7(c), Soman et al. [42]) as a lock-free union-find: a root hi is hooked under lo < hi only by
// CAS(parent[hi], hi, lo), so a link is never overwritten and two vertices that once share a root always do.
// Hence one pass over every arc leaves every arc's endpoints in one tree; pointer jumping then flattens the trees
// to stars whose root is the minimum id (parent[x] < x for every non-root x).  The paper's repeat-until-stable
// loop therefore ends after the first pass.
template <bool HALVE>
__device__ __forceinline__ uint32_t cc_find(uint32_t* parent, uint32_t x) {  // with path halving when HALVE
    uint32_t p = parent[x];
    while (p != x) {
        const uint32_t gp = parent[p];
        if (HALVE && gp != p) parent[x] = gp;  // gp is an ancestor of x: safe under concurrent hooks
        x = p;
        p = gp;
    }
    return x;
}

// HALVE = false (partitioned CC): the only writes to parent are the hooks, so ranks that exchange their hooks keep
// identical parent arrays.  With `pairs`, every successful hook (hi -> lo) is also recorded as a pair (up to cap) for
// the sparse delta exchange; hook_ctr counts all hooks.
template <bool HALVE>
struct CcAppT {
    uint32_t* parent;
    uint32_t* hook_ctr;
    uint32_t* pairs;
    uint32_t cap;
    uint32_t ru;
    __device__ __forceinline__ void begin(uint32_t u) { ru = cc_find<HALVE>(parent, u); }
    __device__ __forceinline__ void end() {}
    __device__ __forceinline__ void vertex(uint32_t) {}
    __device__ __forceinline__ void one(uint32_t v) {
        uint32_t rv = cc_find<HALVE>(parent, v);
        while (ru != rv) {
            const uint32_t hi = max(ru, rv), lo = min(ru, rv);
            if (atomicCAS(parent + hi, hi, lo) == hi) {
                if (hook_ctr) {
                    const uint32_t slot = atomicAdd(hook_ctr, 1u);
                    if (pairs && slot < cap) {
                        pairs[2 * slot] = hi;
                        pairs[2 * slot + 1] = lo;
                    }
                }
                break;
            }
            ru = cc_find<HALVE>(parent, ru);  // hi stopped being a root: re-find both
            rv = cc_find<HALVE>(parent, rv);
        }
    }
    GCGT_MANY_BY_ONE
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for (uint32_t t = 0; t < len; t++) one(s + t);
    }
};
using CcApp = CcAppT<true>;
using CcDistApp = CcAppT<false>;

// Sparse delta merge (partitioned CC): parent[hi] = min(parent[hi], lo) for the received hook pairs.
__global__ void cc_merge_pairs(uint32_t* __restrict__ parent, const uint32_t* __restrict__ pairs, uint64_t npairs) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < npairs; i += (uint64_t)gridDim.x * blockDim.x)
        atomicMin(parent + pairs[2 * i], pairs[2 * i + 1]);
}

}  // namespace gcgt_dev

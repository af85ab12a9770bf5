// contract.cuh — contraction (Alg. 1 l.20-36), the level state kept on the device, the direction
// choice, seeding, CC pointer jumping and the partitioned-BFS helper kernels.
//
// The frontier is a bitmap F plus a queue of its non-zero 32-bit words.  The filter ORs newly discovered vertices
// into the next-frontier bitmap N; the contraction scans N densely: V |= N, F = N, the new vertices' levels are
// written with one coalesced 128-byte store per word, and every non-zero word is appended to the next queue with
// one atomic per warp (the paper's CTA scan + one atomic, at warp granularity).  All per-level bookkeeping (level
// number, queue lengths, direction) lives in device memory, so a level needs no host round trip and the level loop
// can run as a CUDA graph.
#pragma once
#include "device.cuh"

namespace gcgt_dev {

struct LevelState {
    uint32_t dir;       // direction of the level about to run: 0 top-down, 1 bottom-up (BFS)
    uint32_t visited;   // vertices visited so far
    uint32_t nf;        // vertices discovered by the level being committed (commit blocks accumulate)
    uint32_t prev_nf;   // size of the level just expanded
    int32_t level;      // the level being expanded (d); the contraction writes d + 1
    uint32_t qlen[2];   // BFS: queue lengths, ping-pong by level parity
    uint32_t done;      // commit blocks finished (the last one decides)
    uint32_t nonempty;  // levels whose frontier was non-empty
    uint32_t q_off, q_len, q_next;  // BC: current level's range in the all-levels queue, next level's length
    uint32_t ntd, nbu;  // levels run top-down / bottom-up (BFS; kernel-launch accounting of the graph path)
    uint32_t pad;
    unsigned long long mf;  // record bits of the new frontier (dir_bits / dir_edges direction tests)
    unsigned long long mu;  // in-record bits of the vertices visited so far (dir_edges)
};

// Direction choice for the next BFS level (Beamer et al.'s heuristic, on vertex counts): switch to bottom-up when
// the new frontier is large against the unvisited set (nf * alpha > unvisited) and growing, back to top-down when it
// is small against n (nf * beta < n) and shrinking.  With use_bits (symmetric graphs) the top-down -> bottom-up test is Beamer's edge form with CGR bits as
// the work measure: mf * alpha_bits > (unvisited vertices) * (mean record bits).
struct DecideArgs {
    uint64_t n;
    uint32_t alpha10, beta;  // alpha in tenths
    int enabled;
    int use_bits;
    double bits_per_vertex;
    uint32_t alpha_bits10;  // in tenths
    int grow;  // 1: switch to bottom-up only while the frontier grows (Beamer's condition)
    int use_edges;      // Beamer's edge rule with CGR bits as the work measure: mf * alpha > mu
    double mu_total;    // in-CGR bits of all vertices (mu = mu_total - bits of the visited ones)
    uint32_t alpha2_10, guard10;  // second edge test, taken only when the frontier grew by more than guard10 / 10
};

struct CommitArgs {
    uint32_t* __restrict__ V;
    uint32_t* __restrict__ F;      // BFS: rewritten densely; BC: nullptr
    uint32_t* __restrict__ N;
    uint64_t w_lo, w_hi;
    uint32_t* __restrict__ qn;     // next queue (BFS) or the all-levels queue (BC)
    uint32_t* __restrict__ qn_len; // BFS: next queue length
    uint32_t* __restrict__ qcur_len;  // BFS: the consumed queue's length (reset)
    uint32_t* __restrict__ qbits;  // BC: frontier bits per queue entry (all levels)
    uint32_t* __restrict__ lvl_off;  // BC: queue offset of every level
    int32_t* __restrict__ levels;
    LevelState* ls;
    unsigned long long* hub_ctr;   // [2] hub segment / interval chunk queues, reset for the next level
    unsigned long long* cursor;    // the expansion's work cursor [2], reset for the next level
    Offs offs_bits;                // record bits of the new frontier (used when use_mf)
    const uint32_t* __restrict__ wb_out;  // dir_edges: record bits per 32-vertex word, out- and in-CGR (the new
    const uint32_t* __restrict__ wb_in;   // vertices of a word are charged popc/32 of it: one coalesced load)
    int use_mf, use_mu;
    DecideArgs dec;
    int bc;
    int use_cond, use_dcond;
    cudaGraphConditionalHandle cond;   // while-loop condition: the next frontier is non-empty
    cudaGraphConditionalHandle dcond;  // if/else of the next level: 1 = bottom-up
};

__device__ __forceinline__ void decide_body(volatile LevelState* ls, const DecideArgs& d, uint32_t qn_len) {
    if (ls->dir) ls->nbu++;
    else ls->ntd++;
    const uint64_t nf = ls->nf;
    ls->nf = 0;
    const uint64_t visited = (uint64_t)ls->visited + nf;
    ls->visited = (uint32_t)visited;
    const uint64_t nu = d.n - visited, prev = ls->prev_nf;
    uint32_t dir = ls->dir;
    bool to_bu = nf * d.alpha10 > nu * 10;
    if (d.use_bits) to_bu = (double)ls->mf * d.alpha_bits10 > (double)nu * d.bits_per_vertex * 10.0;
    // edge rule (Beamer et al.: m_f > m_u / alpha) with record bits as edge counts: the top-down cost of the next
    // level is the out-record bits of the new frontier, the bottom-up cost at most the in-record bits of the
    // unvisited vertices
    // (r2 sweeps on B200: the vertex-count test suits the web graphs C2/C4; the social and R-MAT graphs gain from
    // the edge test with alpha 25, taken only on explosive frontier growth (nf > guard * previous frontier): there the
    // frontier holds the high-degree vertices -- an expensive top-down level -- and the next level reaches most of
    // the rest, so bottom-up scans stop early; the web graphs' frontiers grow ~1.5x per level at that point)
    if (d.use_edges) {  // in addition to the vertex-count test
        const double mf = (double)ls->mf * 10.0, mu = d.mu_total - (double)ls->mu;
        to_bu = to_bu || mf * d.alpha_bits10 > mu * 100.0 ||
                (mf * d.alpha2_10 > mu * 100.0 && nf * 10 > prev * d.guard10);
    }
    ls->mf = 0;
    if (!d.enabled || nf == 0) dir = 0;
    // (never into bottom-up with a frontier below the bottom-up -> top-down threshold: a whole-graph scan for the
    // last few vertices)
    else if (dir == 0 && to_bu && (nf > prev || !d.grow) && nf * d.beta >= d.n) dir = 1;
    else if (dir == 1 && nf * d.beta < d.n && nf < prev) dir = 0;
    ls->dir = dir;
    ls->prev_nf = (uint32_t)nf;
    if (qn_len) ls->nonempty++;
}

__global__ void __launch_bounds__(kBlock) commit_kernel(CommitArgs a) {
    const volatile LevelState* cls = a.ls;
    const int32_t new_level = cls->level + 1;
    uint32_t qbase = 0;
    if (a.bc) qbase = cls->q_off + cls->q_len;
    const uint32_t lane = lane_id();
    const uint64_t gw = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    uint32_t nf = 0;
    uint64_t mf = 0, mu = 0;
    uint32_t* qlen = a.bc ? &a.ls->q_next : a.qn_len;
    for (uint64_t base = a.w_lo + gw * 32; base < a.w_hi; base += nwarps * 32) {
        const uint64_t w = base + lane;
        uint32_t b = 0;
        if (w < a.w_hi) {
            b = a.N[w];
            if (b) {
                a.N[w] = 0;
                a.V[w] |= b;
            }
            if (a.F && a.F[w] != b) a.F[w] = b;  // F = exactly the new frontier
            if (b && a.use_mu) {
                const uint32_t c = __popc(b);
                mf += ((uint64_t)a.wb_out[w] * c) >> 5;
                mu += ((uint64_t)a.wb_in[w] * c) >> 5;
            }
        }
        nf += __popc(b);
        const uint32_t bal = __ballot_sync(0xffffffffu, b != 0);
        if (bal) {
            uint32_t pos = 0;
            if (lane == 0) pos = atomicAdd(qlen, __popc(bal));
            pos = __shfl_sync(0xffffffffu, pos, 0) + __popc(bal & lanemask_lt());
            if (b) {
                a.qn[qbase + pos] = (uint32_t)w;
                if (a.qbits) a.qbits[qbase + pos] = b;
            }
            for (uint32_t m = bal; m; m &= m - 1) {  // one coalesced 32-id store per new frontier word
                const int j = __ffs(m) - 1;
                const uint32_t bj = __shfl_sync(0xffffffffu, b, j);
                if ((bj >> lane) & 1u) {
                    const uint64_t v = (base + j) * 32 + lane;
                    a.levels[v] = new_level;
                    if (a.use_mf && !a.use_mu) mf += a.offs_bits(v + 1) - a.offs_bits(v);  // coalesced reads
                }
            }
        }
    }
    for (int o = 16; o; o >>= 1) nf += __shfl_xor_sync(0xffffffffu, nf, o);
    if (lane == 0 && nf) atomicAdd(&a.ls->nf, nf);
    if (a.use_mf) {
        for (int o = 16; o; o >>= 1) mf += __shfl_xor_sync(0xffffffffu, mf, o);
        if (lane == 0 && mf) atomicAdd(&a.ls->mf, (unsigned long long)mf);
    }
    if (a.use_mu) {
        for (int o = 16; o; o >>= 1) mu += __shfl_xor_sync(0xffffffffu, mu, o);
        if (lane == 0 && mu) atomicAdd(&a.ls->mu, (unsigned long long)mu);
    }
    // the last block out closes the level: direction, counters, level number, loop condition
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        if (atomicAdd(&a.ls->done, 1u) == gridDim.x - 1) {
            __threadfence();
            volatile LevelState* ls = a.ls;  // other blocks' counts arrived by atomics: read through L2
            ls->done = 0;
            if (a.hub_ctr) {
                a.hub_ctr[0] = 0;
                a.hub_ctr[1] = 0;
            }
            if (a.cursor) {
                a.cursor[0] = 0;
                a.cursor[1] = 0;
            }
            uint32_t next_len;
            if (a.bc) {
                next_len = ls->q_next;
                ls->q_off = qbase;
                ls->q_len = next_len;
                ls->q_next = 0;
                a.lvl_off[new_level + 1] = qbase + next_len;
                ls->nf = 0;
                if (next_len) ls->nonempty++;
            } else {
                next_len = *(volatile uint32_t*)a.qn_len;
                *a.qcur_len = 0;
                decide_body(ls, a.dec, next_len);
            }
            ls->level = new_level;
            if (a.use_cond) {
                cudaGraphSetConditional(a.cond, next_len != 0 ? 1u : 0u);
                if (a.use_dcond) cudaGraphSetConditional(a.dcond, ls->dir);
            }
        }
    }
}

// BFS / BC seed.  The source comes from device memory (written by the host before the launch, so a captured graph
// can be replayed for any source).
__global__ void seed_kernel(const uint32_t* __restrict__ src_p, uint32_t* V, uint32_t* F, uint32_t* q,
                            uint32_t* qbits, int32_t* levels, LevelState* ls, uint32_t* lvl_off, double* sigma) {
    const uint32_t s = *src_p;
    V[s >> 5] = 1u << (s & 31);
    levels[s] = 0;
    if (F) F[s >> 5] = 1u << (s & 31);
    q[0] = s >> 5;
    if (qbits) qbits[0] = 1u << (s & 31);
    if (sigma) sigma[s] = 1.0;
    *ls = LevelState{};
    ls->visited = 1;
    ls->prev_nf = 1;
    ls->qlen[0] = 1;
    ls->q_len = 1;
    if (lvl_off) {
        lvl_off[0] = 0;
        lvl_off[1] = 1;
    }
}

// levels of the vertices the search never reached: -1 (every visited vertex's level was written exactly once, by the
// seed or by the contraction that discovered it, so the levels array needs no initialising pass).
// One thread per 32-vertex word: after a full traversal nearly every word is all-visited, so the pass reads n/8
// bytes and writes almost nothing.
__global__ void finalize_levels(const uint32_t* __restrict__ V, int32_t* __restrict__ levels, uint64_t n) {
    const uint64_t nw = (n + 31) / 32;
    for (uint64_t w = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; w < nw; w += (uint64_t)gridDim.x * blockDim.x) {
        uint32_t unv = ~__ldg(V + w);
        if (n - w * 32 < 32) unv &= (1u << (n - w * 32)) - 1;
        for (; unv; unv &= unv - 1) levels[w * 32 + (__ffs(unv) - 1)] = -1;
    }
}

__global__ void cc_jump(uint32_t* parent, uint64_t n) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n; v += (uint64_t)gridDim.x * blockDim.x) {
        uint32_t x = (uint32_t)v, p = parent[x];
        while (p != x) { x = p; p = parent[x]; }
        parent[v] = x;
    }
}

__global__ void cc_init(uint32_t* parent, uint64_t n) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n; v += (uint64_t)gridDim.x * blockDim.x)
        parent[v] = (uint32_t)v;
}

// BC backward: writes (set) or clears the bitmap words of one level from its queue range (words + frontier bits).
__global__ void bc_level_bits(const uint32_t* __restrict__ q, const uint32_t* __restrict__ qbits, uint32_t len,
                              uint32_t* __restrict__ LB, int set) {
    for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < len; i += gridDim.x * blockDim.x)
        LB[q[i]] = set ? qbits[i] : 0u;
}

// BC backward: X(v) = (1 + delta(v)) / sigma(v) for the vertices of one level (its queue range), once their delta
// is final.
__global__ void bc_level_x(const uint32_t* __restrict__ q, const uint32_t* __restrict__ qbits, uint32_t len,
                           const double* __restrict__ sigma, const double* __restrict__ delta, double* __restrict__ X) {
    for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < len * 32; i += gridDim.x * blockDim.x) {
        const uint32_t e = i >> 5, b = i & 31;
        if ((qbits[e] >> b) & 1u) {
            const uint64_t v = (uint64_t)q[e] * 32 + b;
            X[v] = (1.0 + delta[v]) / sigma[v];
        }
    }
}

// Record bits per 32-vertex word of the owned range [lo, hi) (dir_edges direction rule).
__global__ void word_bits_kernel(Offs offs, uint64_t lo, uint64_t hi, uint32_t* __restrict__ wb) {
    const uint64_t w0 = lo >> 5, nw = ((hi + 31) >> 5) - w0;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < nw; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint64_t a = max((w0 + i) * 32, lo), b = min((w0 + i) * 32 + 32, hi);
        const uint64_t bits = offs(b) - offs(a);
        wb[i] = bits > 0xFFFFFFFFull ? 0xFFFFFFFFu : (uint32_t)bits;
    }
}

__global__ void bswap_words(uint64_t* w, uint64_t n) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x)
        w[i] = __byte_perm((uint32_t)(w[i] >> 32), 0, 0x0123) | ((uint64_t)__byte_perm((uint32_t)w[i], 0, 0x0123) << 32);
}

// ---- partitioned BFS helpers (§8 e) ---------------------------------------------------------------------------------
// Contraction of the owned slice: OR of the P candidate slices received from every rank (plus the owned bottom-up
// finds already in fslice when `keep`), minus visited; writes levels and the owned next-frontier slice; counts new
// vertices into *count.
__global__ void dist_commit(const uint32_t* __restrict__ recv, uint32_t P, uint64_t w_lo, uint64_t nlw,
                            const uint32_t* __restrict__ V, uint32_t* __restrict__ fslice, int32_t* __restrict__ levels,
                            const int32_t* __restrict__ level_p, uint64_t n, unsigned long long* __restrict__ count,
                            int keep) {
    const uint32_t lane = lane_id();
    const int32_t new_level = *level_p + 1;
    uint32_t nf = 0;
    const uint64_t gw = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    for (uint64_t base = gw * 32; base < nlw; base += nwarps * 32) {
        const uint64_t i = base + lane;
        uint32_t b = 0;
        if (i < nlw) {
            b = keep ? fslice[i] : 0u;
            for (uint32_t r = 0; r < P; r++) b |= recv[(uint64_t)r * nlw + i];
            b &= ~V[w_lo + i];
            fslice[i] = b;
        }
        nf += __popc(b);
        for (uint32_t m = __ballot_sync(0xffffffffu, b != 0); m; m &= m - 1) {  // coalesced level stores
            const int j = __ffs(m) - 1;
            const uint32_t bj = __shfl_sync(0xffffffffu, b, j);
            const uint64_t v = (w_lo + base + j) * 32 + lane;
            if (((bj >> lane) & 1u) && v < n) levels[v] = new_level;
        }
    }
    for (int o = 16; o; o >>= 1) nf += __shfl_xor_sync(0xffffffffu, nf, o);
    if (lane == 0 && nf) atomicAdd(count, (unsigned long long)nf);
}

// F = the gathered global frontier; V |= F; counts the frontier (every rank sees the same count, so the
// termination test needs no extra collective) and advances the level.
__global__ void dist_absorb(const uint32_t* __restrict__ Fg, uint32_t* __restrict__ F, uint32_t* __restrict__ V,
                            uint64_t nw, unsigned long long* __restrict__ count) {
    uint32_t c = 0;
    for (uint64_t w = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; w < nw; w += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t b = Fg[w];
        F[w] = b;
        V[w] |= b;
        c += __popc(b);
    }
    for (int o = 16; o; o >>= 1) c += __shfl_xor_sync(0xffffffffu, c, o);
    if (lane_id() == 0 && c) atomicAdd(count, (unsigned long long)c);
}

}  // namespace gcgt_dev

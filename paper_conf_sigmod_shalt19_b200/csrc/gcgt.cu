// gcgt.cu — B200 (sm_100a) device path of GCGT: device residency of the CGR and the traversal kernels.
//
// Pipeline (expansion - filtering - contraction, §6, Fig. 7(a)), re-designed for B200:
//  * Frontier = bitmap F plus a queue of the frontier's non-zero 32-bit words (not a vertex queue): one queue
//    entry per touched word, so contraction costs one atomic per new word instead of one per vertex, and the
//    32 vertices of a word are consecutive ids whose bit offsets / records are contiguous in HBM (BFS-ordered
//    graphs make frontiers clustered).
//  * Filtering tests the visited bitmap V through the read-only path (V is immutable during a level) and claims
//    with atomicOr on the next-frontier bitmap N; an interval run is claimed a word (32 ids) at a time.
//  * A commit step folds N into V / F per level.
//  * Decoding (decode.cuh) is branch-light: 64-bit window + CLZ per codeword.
// Applications: BFS levels (Fig. 7(b)), CC hooking + pointer jumping (Fig. 7(c), Soman [42]), BC forward sigma /
// backward delta (Fig. 7(d), Brandes [9]).
#include <cuda_runtime.h>
#include <cooperative_groups.h>
#include <stdio.h>
#include <string.h>

#include <algorithm>
#include <memory>
#include <string>
#include <vector>

#include "decode.cuh"
#include "internal.h"

namespace cg = cooperative_groups;
using namespace gcgt_dev;

// ------------------------------------------------------------------------------------------------------------------
// errors
// ------------------------------------------------------------------------------------------------------------------
namespace gcgt_internal {
static thread_local std::string g_err;
gcgt_status fail(gcgt_status st, const std::string& msg) {
    g_err = msg;
    return st;
}
void clear_error() { g_err.clear(); }
}  // namespace gcgt_internal
using gcgt_internal::fail;

extern "C" const char* gcgt_last_error(void) { return gcgt_internal::g_err.c_str(); }
extern "C" const char* gcgt_version(void) { return "gcgt-b200 0.1 (sm_100a)"; }

#define CU(call)                                                                                          \
    do {                                                                                                  \
        cudaError_t e_ = (call);                                                                          \
        if (e_ != cudaSuccess) return fail(GCGT_ECUDA, std::string(#call) + ": " + cudaGetErrorString(e_)); \
    } while (0)

// ------------------------------------------------------------------------------------------------------------------
// device graph
// ------------------------------------------------------------------------------------------------------------------
struct Stats {  // device-side counters
    unsigned long long vertices, arcs, bits;
};

struct gcgt_graph {
    int device = 0;
    cudaStream_t stream = nullptr;
    bool own_stream = false;
    uint64_t n = 0, nbits = 0, nw = 0;  // nw = words of an n-bit bitmap
    gcgt_params P{};
    uint64_t lo = 0, hi = 0;
    // CGR
    uint64_t* W = nullptr;     // stream-order words (+2 pad)
    uint64_t* offs = nullptr;  // n + 1
    // work
    uint32_t *V = nullptr, *F = nullptr, *N = nullptr;
    uint32_t* q = nullptr;      // word queue storage (BFS: 2 x nw ping-pong; BC: all levels, nw + n)
    uint32_t* qbits = nullptr;  // BC: frontier bits per queue entry
    uint64_t qcap = 0;
    uint32_t* ctr = nullptr;    // device counters [4]
    Stats* stats = nullptr;
    int32_t* levels = nullptr;
    uint32_t* parent = nullptr;
    double *sigma = nullptr, *delta = nullptr, *bc = nullptr;
    uint32_t* h_ctr = nullptr;  // pinned mirror of ctr
    Stats* h_stats = nullptr;
    cudaEvent_t ev0 = nullptr, ev1 = nullptr;
    int num_sms = 148;
    // profiling of the dominant kernel
    bool profile = false;
    cudaEvent_t kev0 = nullptr, kev1 = nullptr;
    double kernel_ms = 0;
    uint64_t kernel_launches = 0;
};

namespace {

constexpr int kBlock = 256;
constexpr int kWarps = kBlock / 32;

__device__ __forceinline__ uint32_t lane_id() { return threadIdx.x & 31; }

// Appends word index w to the queue; aggregated over the currently converged lanes (one atomic per group).
__device__ __forceinline__ void enqueue_word(uint32_t* __restrict__ qn, uint32_t* __restrict__ qn_len, uint32_t w) {
    cg::coalesced_group g = cg::coalesced_threads();
    uint32_t base = 0;
    if (g.thread_rank() == 0) base = atomicAdd(qn_len, g.size());
    base = g.shfl(base, 0);
    qn[base + g.thread_rank()] = w;
}

__device__ __forceinline__ void add_stats(Stats* st, uint64_t v, uint64_t a, uint64_t b) {
    // warp-reduce then one atomic per warp
    for (int o = 16; o; o >>= 1) {
        v += __shfl_xor_sync(0xffffffffu, v, o);
        a += __shfl_xor_sync(0xffffffffu, a, o);
        b += __shfl_xor_sync(0xffffffffu, b, o);
    }
    if (lane_id() == 0 && v) {
        atomicAdd(&st->vertices, (unsigned long long)v);
        atomicAdd(&st->arcs, (unsigned long long)a);
        atomicAdd(&st->bits, (unsigned long long)b);
    }
}

// ---- frontier iteration -------------------------------------------------------------------------------------------
// Each warp takes `wpb` queue words at a time, expands their set bits into a compact list in shared memory and
// hands one frontier vertex to each lane.  fn(u, lane_active) is called warp-uniformly (lanes without a vertex
// pass active = false), so fn may use warp collectives.
template <class Fn>
__device__ __forceinline__ void for_each_frontier_vertex(const uint32_t* __restrict__ q, uint32_t qlen,
                                                         uint32_t* __restrict__ Fbits, const uint32_t* qbits,
                                                         uint32_t wpb, Fn&& fn) {
    __shared__ uint32_t s_w[kWarps][32], s_b[kWarps][32], s_pre[kWarps][33];
    const uint32_t wid = threadIdx.x >> 5, lane = lane_id();
    const uint64_t gw = (uint64_t)blockIdx.x * kWarps + wid, nwarps = (uint64_t)gridDim.x * kWarps;
    for (uint64_t base = gw * wpb; base < qlen; base += nwarps * wpb) {
        uint32_t w = 0, bits = 0;
        if (lane < wpb && base + lane < qlen) {
            w = q[base + lane];
            if (qbits) bits = qbits[base + lane];
            else { bits = Fbits[w]; Fbits[w] = 0; }
        }
        const uint32_t c = __popc(bits);
        uint32_t incl = c;
        for (int o = 1; o < 32; o <<= 1) {
            const uint32_t t = __shfl_up_sync(0xffffffffu, incl, o);
            if (lane >= (uint32_t)o) incl += t;
        }
        s_w[wid][lane] = w;
        s_b[wid][lane] = bits;
        s_pre[wid][lane + 1] = incl;
        if (lane == 0) s_pre[wid][0] = 0;
        __syncwarp();
        const uint32_t total = s_pre[wid][32];
        for (uint32_t t = 0; t < total; t += 32) {
            const uint32_t j = t + lane;
            uint32_t u = 0;
            const bool act = j < total;
            if (act) {
                uint32_t lo = 0, hi = 31;  // owner: largest o with s_pre[o] <= j
                while (lo < hi) {
                    const uint32_t mid = (lo + hi + 1) >> 1;
                    if (s_pre[wid][mid] <= j) lo = mid; else hi = mid - 1;
                }
                const uint32_t r = j - s_pre[wid][lo];
                const uint32_t pos = __fns(s_b[wid][lo], 0, (int)r + 1);
                u = s_w[wid][lo] * 32 + pos;
            }
            fn(u, act);
        }
        __syncwarp();
    }
}

// ---- BFS ------------------------------------------------------------------------------------------------------------
struct BfsVisitor {
    const uint32_t* __restrict__ V;
    uint32_t* __restrict__ N;
    uint32_t* __restrict__ qn;
    uint32_t* __restrict__ qn_len;
    __device__ __forceinline__ void claim(uint32_t w, uint32_t mask) {
        const uint32_t cand = mask & ~__ldg(V + w);
        if (!cand) return;
        const uint32_t old = atomicOr(N + w, cand);
        if (old == 0) enqueue_word(qn, qn_len, w);
    }
    __device__ __forceinline__ void one(uint32_t v) { claim(v >> 5, 1u << (v & 31)); }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {  // interval: one claim per 32-id word
        uint32_t e = s + len;                                           // exclusive
        while (s < e) {
            const uint32_t w = s >> 5, b0 = s & 31;
            const uint32_t nb = min(32u - b0, e - s);
            const uint32_t mask = (nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0;
            claim(w, mask);
            s += nb;
        }
    }
};

template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock) bfs_expand(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                                     uint32_t min_len, uint32_t seg_bits, int32_t level,
                                                     const uint32_t* __restrict__ q, const uint32_t* __restrict__ qlen_p,
                                                     uint32_t* __restrict__ F, const uint32_t* __restrict__ V,
                                                     uint32_t* __restrict__ N, uint32_t* __restrict__ qn,
                                                     uint32_t* __restrict__ qn_len, int32_t* __restrict__ levels,
                                                     uint32_t wpb, Stats* st) {
    const uint32_t qlen = *qlen_p;
    BfsVisitor vis{V, N, qn, qn_len};
    uint64_t nv = 0, na = 0, nb = 0;
    for_each_frontier_vertex(q, qlen, F, nullptr, wpb, [&](uint32_t u, bool act) {
        if (!act) return;
        levels[u] = level;
        const uint64_t p0 = ldg64(offs + u), p1 = ldg64(offs + u + 1);
        na += walk_record<K, SEG>(W, p0, u, min_len, seg_bits, vis);
        nv += 1;
        nb += p1 - p0;
    });
    add_stats(st, nv, na, nb);
}

// Folds the next frontier into V and F: for every queued word, V |= N, F = N, N = 0.
__global__ void bfs_commit(const uint32_t* __restrict__ qn, const uint32_t* __restrict__ qn_len,
                           uint32_t* __restrict__ V, uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                           uint32_t* __restrict__ qbits_out, uint32_t* __restrict__ reset_ctr) {
    const uint32_t len = *qn_len;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < len; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t w = qn[i];
        const uint32_t b = N[w];
        N[w] = 0;
        V[w] |= b;
        if (qbits_out) qbits_out[i] = b;
        else F[w] = b;
    }
    if (reset_ctr && blockIdx.x == 0 && threadIdx.x == 0) *reset_ctr = 0;
}

__global__ void bfs_seed(uint32_t s, uint32_t* V, uint32_t* F, uint32_t* q, uint32_t* qlen, uint32_t* qbits) {
    V[s >> 5] = 1u << (s & 31);
    if (F) F[s >> 5] = 1u << (s & 31);
    q[0] = s >> 5;
    if (qbits) qbits[0] = 1u << (s & 31);
    *qlen = 1;
}

__global__ void bswap_words(uint64_t* w, uint64_t n) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x)
        w[i] = __byte_perm((uint32_t)(w[i] >> 32), 0, 0x0123) | ((uint64_t)__byte_perm((uint32_t)w[i], 0, 0x0123) << 32);
}

// ---- CC -------------------------------------------------------------------------------------------------------------
// Hooking (Fig. 7(c), Soman et al. [42]) as a lock-free union-find: a root hi is hooked under lo < hi only by
// CAS(parent[hi], hi, lo), so a link is never overwritten and two vertices that once share a root always do.
// Hence one pass over every arc leaves every arc's endpoints in one tree; pointer jumping then flattens the trees
// to stars whose root is the minimum id (parent[x] < x for every non-root x).  The paper's repeat-until-stable
// loop therefore ends after the first pass.
__device__ __forceinline__ uint32_t cc_find(uint32_t* parent, uint32_t x) {  // with path halving
    uint32_t p = parent[x];
    while (p != x) {
        const uint32_t gp = parent[p];
        if (gp != p) parent[x] = gp;  // gp is an ancestor of x: safe under concurrent hooks
        x = p;
        p = gp;
    }
    return x;
}

struct CcVisitor {
    uint32_t* parent;
    uint32_t ru;
    uint32_t hooks;
    __device__ __forceinline__ void one(uint32_t v) {
        uint32_t rv = cc_find(parent, v);
        while (ru != rv) {
            const uint32_t hi = max(ru, rv), lo = min(ru, rv);
            if (atomicCAS(parent + hi, hi, lo) == hi) { hooks++; break; }
            ru = cc_find(parent, ru);  // hi stopped being a root: re-find both
            rv = cc_find(parent, rv);
        }
    }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for (uint32_t t = 0; t < len; t++) one(s + t);
    }
};

template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock) cc_hook(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                                  uint32_t min_len, uint32_t seg_bits, uint64_t lo, uint64_t hi,
                                                  uint32_t* parent, uint32_t* hooks, Stats* st) {
    uint64_t nv = 0, na = 0, nb = 0, nh = 0;
    for (uint64_t u = lo + (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; u < hi;
         u += (uint64_t)gridDim.x * blockDim.x) {
        CcVisitor vis{parent, cc_find(parent, (uint32_t)u), 0};
        const uint64_t p0 = ldg64(offs + u), p1 = ldg64(offs + u + 1);
        na += walk_record<K, SEG>(W, p0, u, min_len, seg_bits, vis);
        nv++;
        nb += p1 - p0;
        nh += vis.hooks;
    }
    add_stats(st, nv, na, nb);
    for (int o = 16; o; o >>= 1) nh += __shfl_xor_sync(0xffffffffu, nh, o);
    if (lane_id() == 0 && nh) atomicAdd(hooks, (uint32_t)nh);
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

// ---- BC -------------------------------------------------------------------------------------------------------------
struct BcFwdVisitor {
    const uint32_t* __restrict__ V;
    uint32_t* __restrict__ N;
    uint32_t* __restrict__ qn;
    uint32_t* __restrict__ qn_len;
    double* sigma;
    double su;
    __device__ __forceinline__ void claim(uint32_t w, uint32_t mask) {
        const uint32_t cand = mask & ~__ldg(V + w);  // not at level <= d: level(v) = d + 1
        if (!cand) return;
        const uint32_t old = atomicOr(N + w, cand);
        if (old == 0) enqueue_word(qn, qn_len, w);
        uint32_t c = cand;
        while (c) {
            const int b = __ffs(c) - 1;
            c &= c - 1;
            atomicAdd(sigma + (uint64_t)w * 32 + b, su);
        }
    }
    __device__ __forceinline__ void one(uint32_t v) { claim(v >> 5, 1u << (v & 31)); }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        uint32_t e = s + len;
        while (s < e) {
            const uint32_t w = s >> 5, b0 = s & 31;
            const uint32_t nb = min(32u - b0, e - s);
            claim(w, (nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0);
            s += nb;
        }
    }
};

template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock) bc_forward(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                                     uint32_t min_len, uint32_t seg_bits, int32_t level,
                                                     const uint32_t* __restrict__ q, const uint32_t* __restrict__ qbits,
                                                     const uint32_t* __restrict__ qlen_p, const uint32_t* __restrict__ V,
                                                     uint32_t* __restrict__ N, uint32_t* __restrict__ qn,
                                                     uint32_t* __restrict__ qn_len, int32_t* __restrict__ levels,
                                                     double* sigma, uint32_t wpb, Stats* st) {
    const uint32_t qlen = *qlen_p;
    uint64_t nv = 0, na = 0, nb = 0;
    for_each_frontier_vertex(q, qlen, nullptr, qbits, wpb, [&](uint32_t u, bool act) {
        if (!act) return;
        levels[u] = level;
        BcFwdVisitor vis{V, N, qn, qn_len, sigma, sigma[u]};
        const uint64_t p0 = ldg64(offs + u), p1 = ldg64(offs + u + 1);
        na += walk_record<K, SEG>(W, p0, u, min_len, seg_bits, vis);
        nv++;
        nb += p1 - p0;
    });
    add_stats(st, nv, na, nb);
}

struct BcBwdVisitor {
    const int32_t* __restrict__ levels;
    const double* __restrict__ sigma;
    const double* __restrict__ delta;
    int32_t next;
    double sv;
    double acc;
    __device__ __forceinline__ void one(uint32_t w) {
        if (levels[w] == next) acc += sv / sigma[w] * (1.0 + delta[w]);
    }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for (uint32_t t = 0; t < len; t++) one(s + t);
    }
};

// delta(v) = sum_{w in out(v), d(w) = d(v)+1} sigma(v)/sigma(w) (1 + delta(w))  (Fig. 7(d), pull form)
template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock) bc_backward(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                                      uint32_t min_len, uint32_t seg_bits, int32_t level,
                                                      const uint32_t* __restrict__ q, const uint32_t* __restrict__ qbits,
                                                      uint32_t qlen, uint32_t source, const int32_t* __restrict__ levels,
                                                      const double* __restrict__ sigma, double* __restrict__ delta,
                                                      double* __restrict__ bc, uint32_t wpb, Stats* st) {
    uint64_t nv = 0, na = 0, nb = 0;
    for_each_frontier_vertex(q, qlen, nullptr, qbits, wpb, [&](uint32_t v, bool act) {
        if (!act) return;
        BcBwdVisitor vis{levels, sigma, delta, level + 1, sigma[v], 0.0};
        const uint64_t p0 = ldg64(offs + v), p1 = ldg64(offs + v + 1);
        na += walk_record<K, SEG>(W, p0, v, min_len, seg_bits, vis);
        const double d = vis.acc;
        delta[v] = d;
        if (v != source) bc[v] += d;
        nv++;
        nb += p1 - p0;
    });
    add_stats(st, nv, na, nb);
}

// ---- dispatch -------------------------------------------------------------------------------------------------------
#define GCGT_DISPATCH(P, KERNEL, GRID, BLOCK, STREAM, ...)                                                      \
    do {                                                                                                        \
        const bool seg_ = (P).residual_segment_len != 0;                                                        \
        switch ((P).zeta_k) {                                                                                   \
            case 1: if (seg_) KERNEL<1, true><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__);                         \
                    else KERNEL<1, false><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__); break;                      \
            case 2: if (seg_) KERNEL<2, true><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__);                         \
                    else KERNEL<2, false><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__); break;                      \
            case 3: if (seg_) KERNEL<3, true><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__);                         \
                    else KERNEL<3, false><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__); break;                      \
            case 4: if (seg_) KERNEL<4, true><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__);                         \
                    else KERNEL<4, false><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__); break;                      \
            default: if (seg_) KERNEL<5, true><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__);                        \
                    else KERNEL<5, false><<<GRID, BLOCK, 0, STREAM>>>(__VA_ARGS__); break;                      \
        }                                                                                                       \
    } while (0)

// Grid for a frontier of qlen words: aim for ~1 word per lane when the queue is small, batches of 32 otherwise.
inline void frontier_launch(const gcgt_graph* g, uint32_t qlen, int* grid, uint32_t* wpb) {
    const uint64_t max_warps = (uint64_t)g->num_sms * 2048 / 32;  // one wave at full occupancy
    uint32_t b = 1;
    while (b < 32 && (uint64_t)qlen > max_warps * b) b <<= 1;
    uint64_t warps = ((uint64_t)qlen + b - 1) / b;
    uint64_t blocks = std::max<uint64_t>(1, (warps + kWarps - 1) / kWarps);
    *grid = (int)std::min<uint64_t>(blocks, (uint64_t)g->num_sms * 8);
    *wpb = b;
}

inline int flat_grid(const gcgt_graph* g, uint64_t n) {
    return (int)std::max<uint64_t>(1, std::min<uint64_t>((n + kBlock - 1) / kBlock, (uint64_t)g->num_sms * 16));
}

gcgt_status copy_out(gcgt_graph* g, void* dst, const void* src, size_t bytes, int placement) {
    CU(cudaMemcpyAsync(dst, src, bytes, placement == GCGT_OUT_DEVICE ? cudaMemcpyDeviceToDevice : cudaMemcpyDeviceToHost,
                       g->stream));
    return GCGT_OK;
}

// Brackets one launch of the dominant kernel when profiling (the caller syncs before reading).
inline gcgt_status kprof_begin(gcgt_graph* g) {
    if (g->profile) CU(cudaEventRecord(g->kev0, g->stream));
    return GCGT_OK;
}
inline gcgt_status kprof_end(gcgt_graph* g) {
    if (g->profile) CU(cudaEventRecord(g->kev1, g->stream));
    return GCGT_OK;
}
inline gcgt_status kprof_collect(gcgt_graph* g) {  // after a stream sync
    if (!g->profile) return GCGT_OK;
    float ms = 0;
    CU(cudaEventElapsedTime(&ms, g->kev0, g->kev1));
    g->kernel_ms += ms;
    g->kernel_launches++;
    return GCGT_OK;
}

gcgt_status begin_call(gcgt_graph* g) {
    gcgt_internal::clear_error();
    CU(cudaSetDevice(g->device));
    g->kernel_ms = 0;
    g->kernel_launches = 0;
    CU(cudaMemsetAsync(g->stats, 0, sizeof(Stats), g->stream));
    CU(cudaEventRecord(g->ev0, g->stream));
    return GCGT_OK;
}

gcgt_status end_call(gcgt_graph* g, gcgt_stats* out, uint32_t iterations) {
    CU(cudaEventRecord(g->ev1, g->stream));
    CU(cudaMemcpyAsync(g->h_stats, g->stats, sizeof(Stats), cudaMemcpyDeviceToHost, g->stream));
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
    if (out) {
        float ms = 0;
        CU(cudaEventElapsedTime(&ms, g->ev0, g->ev1));
        out->iterations = iterations;
        out->reserved = 0;
        out->vertices_expanded = g->h_stats->vertices;
        out->arcs_decoded = g->h_stats->arcs;
        out->cgr_bits_decoded = g->h_stats->bits;
        out->device_ms = ms;
        out->kernel_ms = g->kernel_ms;
        out->kernel_launches = g->kernel_launches;
    }
    return GCGT_OK;
}

template <class T>
gcgt_status dalloc(T** p, uint64_t count) {
    cudaError_t e = cudaMalloc((void**)p, std::max<uint64_t>(1, count) * sizeof(T));
    if (e != cudaSuccess) return fail(GCGT_ENOMEM, std::string("cudaMalloc: ") + cudaGetErrorString(e));
    return GCGT_OK;
}

}  // namespace

// ------------------------------------------------------------------------------------------------------------------
// C ABI
// ------------------------------------------------------------------------------------------------------------------
extern "C" void gcgt_unload(gcgt_graph* g) {
    if (!g) return;
    cudaSetDevice(g->device);
    if (g->stream) cudaStreamSynchronize(g->stream);
    cudaFree(g->W); cudaFree(g->offs); cudaFree(g->V); cudaFree(g->F); cudaFree(g->N); cudaFree(g->q);
    cudaFree(g->qbits); cudaFree(g->ctr); cudaFree(g->stats); cudaFree(g->levels); cudaFree(g->parent);
    cudaFree(g->sigma); cudaFree(g->delta); cudaFree(g->bc);
    if (g->h_ctr) cudaFreeHost(g->h_ctr);
    if (g->h_stats) cudaFreeHost(g->h_stats);
    if (g->ev0) cudaEventDestroy(g->ev0);
    if (g->ev1) cudaEventDestroy(g->ev1);
    if (g->kev0) cudaEventDestroy(g->kev0);
    if (g->kev1) cudaEventDestroy(g->kev1);
    if (g->own_stream && g->stream) cudaStreamDestroy(g->stream);
    delete g;
}

extern "C" gcgt_status gcgt_load(const gcgt_cgr* c, const gcgt_load_opts* opts, gcgt_graph** out) {
    gcgt_internal::clear_error();
    if (!c || !out) return fail(GCGT_EINVAL, "null argument");
    gcgt_load_opts o{};
    if (opts) o = *opts;
    if (o.nranks > 1) return fail(GCGT_EINVAL, "multi-rank load: use gcgt_load with the NCCL build (not in this build)");
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev == 0) return fail(GCGT_ECUDA, "no CUDA device");
    if (o.device < 0 || o.device >= ndev) return fail(GCGT_EINVAL, "bad device ordinal");
    std::unique_ptr<gcgt_graph, void (*)(gcgt_graph*)> g(new gcgt_graph(), gcgt_unload);
    g->device = o.device;
    CU(cudaSetDevice(o.device));
    cudaDeviceProp prop;
    CU(cudaGetDeviceProperties(&prop, o.device));
    g->num_sms = prop.multiProcessorCount;
    if (o.stream) g->stream = (cudaStream_t)o.stream;
    else {
        CU(cudaStreamCreateWithFlags(&g->stream, cudaStreamNonBlocking));
        g->own_stream = true;
    }
    g->n = c->n;
    g->nbits = c->nbits;
    g->P = c->params;
    g->lo = 0;
    g->hi = c->n;
    g->nw = (c->n + 31) / 32 + 1;
    const uint64_t nwords = (c->nbits + 63) / 64 + 2;
    gcgt_status st;
    if ((st = dalloc(&g->W, nwords)) || (st = dalloc(&g->offs, g->n + 1)) || (st = dalloc(&g->V, g->nw)) ||
        (st = dalloc(&g->F, g->nw)) || (st = dalloc(&g->N, g->nw)) || (st = dalloc(&g->ctr, 8)) ||
        (st = dalloc(&g->stats, 1)) || (st = dalloc(&g->levels, g->n)))
        return st;
    g->qcap = 2 * g->nw;
    if ((st = dalloc(&g->q, g->qcap))) return st;
    CU(cudaMallocHost((void**)&g->h_ctr, 8 * sizeof(uint32_t)));
    CU(cudaMallocHost((void**)&g->h_stats, sizeof(Stats)));
    CU(cudaEventCreate(&g->ev0));
    CU(cudaEventCreate(&g->ev1));
    CU(cudaEventCreate(&g->kev0));
    CU(cudaEventCreate(&g->kev1));
    CU(cudaMemcpyAsync(g->W, c->words.data(), nwords * sizeof(uint64_t), cudaMemcpyHostToDevice, g->stream));
    CU(cudaMemcpyAsync(g->offs, c->bit_offsets.data(), (g->n + 1) * sizeof(uint64_t), cudaMemcpyHostToDevice,
                       g->stream));
    bswap_words<<<flat_grid(g.get(), nwords), kBlock, 0, g->stream>>>(g->W, nwords);
    CU(cudaMemsetAsync(g->N, 0, g->nw * 4, g->stream));
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
    *out = g.release();
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_profile(gcgt_graph* g, int enable) {
    if (!g) return fail(GCGT_EINVAL, "null graph");
    g->profile = enable != 0;
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_graph_range(const gcgt_graph* g, uint64_t* lo, uint64_t* hi) {
    if (!g) return fail(GCGT_EINVAL, "null graph");
    if (lo) *lo = g->lo;
    if (hi) *hi = g->hi;
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_bfs(gcgt_graph* g, uint32_t source, int32_t* levels, int placement, gcgt_stats* stats) {
    if (!g || !levels) return fail(GCGT_EINVAL, "null argument");
    if (source >= g->n) return fail(GCGT_ERANGE, "source >= n");
    gcgt_status st;
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->F, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
    CU(cudaMemsetAsync(g->ctr, 0, 8 * 4, s));
    uint32_t* q[2] = {g->q, g->q + g->nw};
    bfs_seed<<<1, 1, 0, s>>>(source, g->V, g->F, q[0], g->ctr + 0, nullptr);
    const uint32_t seg_bits = 8 * g->P.residual_segment_len;
    uint32_t qlen = 1, level = 0;
    while (qlen) {
        const int cur = level & 1, nxt = cur ^ 1;
        int grid;
        uint32_t wpb;
        frontier_launch(g, qlen, &grid, &wpb);
        if ((st = kprof_begin(g))) return st;
        GCGT_DISPATCH(g->P, bfs_expand, grid, kBlock, s, g->W, g->offs, g->P.min_interval_len, seg_bits,
                      (int32_t)level, q[cur], g->ctr + cur, g->F, g->V, g->N, q[nxt], g->ctr + nxt, g->levels, wpb,
                      g->stats);
        if ((st = kprof_end(g))) return st;
        bfs_commit<<<flat_grid(g, g->nw), kBlock, 0, s>>>(q[nxt], g->ctr + nxt, g->V, g->F, g->N, nullptr,
                                                           g->ctr + cur);
        CU(cudaMemcpyAsync(g->h_ctr + nxt, g->ctr + nxt, 4, cudaMemcpyDeviceToHost, s));
        CU(cudaStreamSynchronize(s));
        if ((st = kprof_collect(g))) return st;
        qlen = g->h_ctr[nxt];
        level++;
    }
    if ((st = copy_out(g, levels, g->levels, g->n * 4, placement))) return st;
    return end_call(g, stats, level);
}

extern "C" gcgt_status gcgt_cc(gcgt_graph* g, uint32_t* labels, int placement, gcgt_stats* stats) {
    if (!g || !labels) return fail(GCGT_EINVAL, "null argument");
    gcgt_status st;
    if (!g->parent && (st = dalloc(&g->parent, g->n))) return st;
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    const uint32_t seg_bits = 8 * g->P.residual_segment_len;
    cc_init<<<flat_grid(g, g->n), kBlock, 0, s>>>(g->parent, g->n);
    CU(cudaMemsetAsync(g->ctr, 0, 4, s));
    if ((st = kprof_begin(g))) return st;
    GCGT_DISPATCH(g->P, cc_hook, flat_grid(g, g->n), kBlock, s, g->W, g->offs, g->P.min_interval_len, seg_bits,
                  (uint64_t)0, g->n, g->parent, g->ctr, g->stats);
    if ((st = kprof_end(g))) return st;
    cc_jump<<<flat_grid(g, g->n), kBlock, 0, s>>>(g->parent, g->n);
    if ((st = copy_out(g, labels, g->parent, g->n * 4, placement))) return st;
    CU(cudaStreamSynchronize(s));
    if ((st = kprof_collect(g))) return st;
    return end_call(g, stats, 1);
}

extern "C" gcgt_status gcgt_bc(gcgt_graph* g, const uint32_t* sources, uint32_t k, double* bc, int placement,
                               gcgt_stats* stats) {
    if (!g || !bc || (k && !sources)) return fail(GCGT_EINVAL, "null argument");
    for (uint32_t i = 0; i < k; i++)
        if (sources[i] >= g->n) return fail(GCGT_ERANGE, "source >= n");
    gcgt_status st;
    if (!g->sigma) {
        if ((st = dalloc(&g->sigma, g->n)) || (st = dalloc(&g->delta, g->n)) || (st = dalloc(&g->bc, g->n)) ||
            (st = dalloc(&g->qbits, g->n + g->nw)))
            return st;
        uint32_t* bigq = nullptr;
        if ((st = dalloc(&bigq, g->n + g->nw))) return st;
        cudaFree(g->q);
        g->q = bigq;
        g->qcap = g->n + g->nw;
    }
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    const uint32_t seg_bits = 8 * g->P.residual_segment_len;
    CU(cudaMemsetAsync(g->bc, 0, g->n * 8, s));
    std::vector<uint32_t> lvl_off;
    for (uint32_t si = 0; si < k; si++) {
        const uint32_t src = sources[si];
        CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
        CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
        CU(cudaMemsetAsync(g->sigma, 0, g->n * 8, s));
        CU(cudaMemsetAsync(g->ctr, 0, 8 * 4, s));
        double one = 1.0;
        CU(cudaMemcpyAsync(g->sigma + src, &one, 8, cudaMemcpyHostToDevice, s));
        // level d occupies q[lvl_off[d] .. lvl_off[d+1]); ctr[0] = running total of queued words
        bfs_seed<<<1, 1, 0, s>>>(src, g->V, nullptr, g->q, g->ctr + 0, g->qbits);
        lvl_off.assign(1, 0);
        uint32_t total = 1, level = 0;
        // ctr[1] = length of the level being built; the kernels index q from lvl_off
        while (true) {
            const uint32_t off = lvl_off.back(), qlen = total - off;
            lvl_off.push_back(total);
            if (!qlen) break;
            CU(cudaMemcpyAsync(g->ctr + 2, &qlen, 4, cudaMemcpyHostToDevice, s));
            CU(cudaMemsetAsync(g->ctr + 1, 0, 4, s));
            int grid;
            uint32_t wpb;
            frontier_launch(g, qlen, &grid, &wpb);
            if ((st = kprof_begin(g))) return st;
            GCGT_DISPATCH(g->P, bc_forward, grid, kBlock, s, g->W, g->offs, g->P.min_interval_len, seg_bits,
                          (int32_t)level, g->q + off, g->qbits + off, g->ctr + 2, g->V, g->N, g->q + total,
                          g->ctr + 1, g->levels, g->sigma, wpb, g->stats);
            if ((st = kprof_end(g))) return st;
            bfs_commit<<<flat_grid(g, g->nw), kBlock, 0, s>>>(g->q + total, g->ctr + 1, g->V, nullptr, g->N,
                                                               g->qbits + total, nullptr);
            CU(cudaMemcpyAsync(g->h_ctr + 1, g->ctr + 1, 4, cudaMemcpyDeviceToHost, s));
            CU(cudaStreamSynchronize(s));
            if ((st = kprof_collect(g))) return st;
            total += g->h_ctr[1];
            level++;
        }
        // lvl_off has D+2 entries: levels 0..D-1 plus the empty terminator
        const int D = (int)lvl_off.size() - 2;
        for (int d = D - 1; d >= 0; d--) {
            const uint32_t off = lvl_off[d], qlen = lvl_off[d + 1] - off;
            int grid;
            uint32_t wpb;
            frontier_launch(g, qlen, &grid, &wpb);
            GCGT_DISPATCH(g->P, bc_backward, grid, kBlock, s, g->W, g->offs, g->P.min_interval_len, seg_bits,
                          (int32_t)d, g->q + off, g->qbits + off, qlen, src, g->levels, g->sigma, g->delta, g->bc, wpb,
                          g->stats);
        }
    }
    if ((st = copy_out(g, bc, g->bc, g->n * 8, placement))) return st;
    return end_call(g, stats, k);
}

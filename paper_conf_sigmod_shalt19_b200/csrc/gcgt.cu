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
#include <cooperative_groups/reduce.h>
#include <cub/cub.cuh>
#include <stdio.h>
#include <string.h>

#include <algorithm>
#include <chrono>
#include <memory>
#include <mutex>
#include <string>
#include <type_traits>
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

struct HubEntry {
    uint64_t base;     // bit position of the vertex's first residual segment
    uint32_t u;        // vertex
    uint32_t seg_off;  // first flattened segment index of this entry (entries are ordered by seg_off)
    uint32_t epoch;    // expansion launch that published the entry (fused hub consumption waits for it)
    uint32_t pad;
};

// A long interval (more than long_len ids) deferred to the level's long-range queue and expanded grid-wide in chunks
// of lr_chunk ids: the Two-Phase Traversal's "long interval expanded by the whole thread group" (Alg. 2 l.23-32,
// PAPER.md:667-688) at grid scale.  Entries are ordered by chunk_off (one packed atomic hands out both indices).
struct LongRange {
    uint32_t u, start, len, chunk_off;
    uint32_t epoch;  // as HubEntry::epoch
};

struct HeavyEntry {
    uint64_t p;    // first bit after the itvNum field
    uint32_t u;
    uint32_t itv;  // interval count
    uint64_t deg;  // unsegmented records: degree (else 0)
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
    uint64_t* offs = nullptr;        // offs[u] for owned u in [lo, hi] (points offs_alloc - lo)
    uint64_t* offs_alloc = nullptr;  // hi - lo + 1 re-based offsets
    int rank = 0, nranks = 1;
    uint64_t* inW = nullptr;     // in-CGR (transpose) for bottom-up; aliases W / offs when symmetric
    uint64_t* inOffs = nullptr;
    bool in_owned = false;       // inW / inOffs are separate allocations
    // host-resident CGR (§8 f4, gcgt_load_opts.host_resident): W / inW point into pinned, mapped host memory that
    // the kernels read over the host link (zero copy); only O(n) tables live in HBM
    uint64_t* hostW = nullptr;
    uint64_t* hostInW = nullptr;
    bool dir_opt = false;        // direction-optimizing BFS enabled (in-CGR available)
    // interval checkpoint table (derived at load) + per-level chunk queue
    uint32_t hv_n = 0, ck_c = 4;
    uint32_t *hv_ids = nullptr, *hv_ptr = nullptr, *hv_rem = nullptr, *ck_prev = nullptr;
    uint32_t *hv_wptr = nullptr, *hv_bits = nullptr;  // per-word index of hv_ids (hv_index)
    uint64_t *hv_after = nullptr, *ck_pos = nullptr;
    LongRange* lrq = nullptr;              // per-level long-range queue
    unsigned long long* lr_ctr = nullptr;  // (entries << 32) | chunks
    uint32_t long_len = 1024, lr_chunk = 256;
    // uncompressed baseline (gcgt_load_csr, §8 f3): device CSR (+ in-lists for bottom-up) instead of the CGR
    bool is_csr = false;
    uint64_t* crow = nullptr;
    uint32_t* ccol = nullptr;
    uint64_t* crow_in = nullptr;
    uint32_t* ccol_in = nullptr;
    bool csr_in_owned = false;
    void* csr_hubq = nullptr;
    unsigned long long* mf = nullptr;  // record bits (CSR: arcs) of the new frontier, for bfs_decide
    // direction test: record bits (Beamer's edge form) on symmetric graphs, vertex counts on directed ones (sweep of
    // round 1: R-MAT 1.39 -> 0.60 ms with bits; the directed web / social recipes are faster with vertex counts)
    bool dir_bits = false;
    uint32_t alpha_bits = 30;
    uint32_t* bstate = nullptr;  // BFS direction state [8]: 0 dir (0 TD, 1 BU), 1 visited, 2 new-frontier count,
                                 // 3 previous frontier count
    // work
    uint32_t *V = nullptr, *F = nullptr, *N = nullptr;
    uint32_t* q = nullptr;      // word queue storage (BFS: 2 x nw ping-pong; BC: all levels, nw + n)
    uint32_t* qbits = nullptr;  // BC: frontier bits per queue entry
    uint64_t qcap = 0;
    uint32_t* ctr = nullptr;    // device counters [8]
    HubEntry* hubq = nullptr;   // per-level hub queue (capacity = hub vertices + 1)
    unsigned long long* cursor = nullptr;  // [0] work cursor, [1] finished-warp count (expand_kernel)
    HeavyEntry* heavyq = nullptr;          // per-level heavy-vertex queue (capacity = heavy vertices + 1)
    // tuning knobs (defaults; GCGT_TUNE="staged=0,heavy_itv=16,hub_segs=8,wpb_max=8" overrides at load)
    // defaults from the C2 sweep (profiles/r1_sweep_c2.txt): per-codeword window reads beat register staging, and
    // deferring long interval areas to a separate pass costs more than the in-batch straggler it removes
    bool staged = false;
    bool persistent = false;
    uint32_t chunk = 4;       // BFS levels enqueued per host check of the queue length (GCGT_TUNE chunk=N)
    uint32_t nfilter = 0;     // BfsApp: filter claims on an L1 read of N before the atomic (GCGT_TUNE nfilter=1)
    uint32_t flatb = 0;       // phase B lane-refill loop (GCGT_TUNE flatb=1; measured no faster on C2, session 3)
    uint32_t fuse_warps = 0;  // fused hub consumption: consumer warps per expand block (GCGT_TUNE fuse=N; 0 = hub_kernel)
    bool dir_opt_knob = true;
    uint32_t engine = 0;  // 0 = phase kernel; 1 = state-machine kernel (measured slower on C2: lone long tasks)  // BFS: all levels in one cooperative launch (measured slower on C2; GCGT_TUNE knob)
    uint32_t heavy_itv = 0xFFFFFFFFu, heavy_res = 1024, hub_segs = 8, wpb_max = 8;
    uint32_t bu_kernel = 1;  // bottom-up kernel: 1 = per-word (lane = vertex id), 2 = compacted chunks (bu_words/bu_batch)
    uint32_t bu_words = 8, bu_batch = 4;  // bottom-up: frontier words per warp chunk, residuals per probe batch
    uint32_t bu_alpha = 4, bu_beta = 128;  // switch thresholds on vertex counts (beta: r1 session-4 sweep, C2+C3)
    uint32_t* heavy_len = nullptr;
    unsigned long long* hub_ctr = nullptr;
    uint32_t* fuse_ctr = nullptr;  // fused hub consumption counters [4] (Ctx::fuse_ctr)
    unsigned long long* bu_cur = nullptr;  // bu_kernel chunk cursor [2]
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
    static constexpr int kKev = 64;           // event pairs: one per profiled launch between host syncs
    cudaEvent_t kevp[2 * kKev] = {};
    int kev_n = 0;
    bool spans = false;  // per-level span events (profile mode 2): the level loop then waits per level
    cudaEvent_t sev[5] = {nullptr, nullptr, nullptr, nullptr, nullptr};  // span marks within a BFS level
    double span_ms[4] = {0, 0, 0, 0};  // expand(+heavy), hub, bottom-up, contraction (+decide)
    double kernel_ms = 0;
    uint64_t kernel_launches = 0;
    uint64_t launches = 0;  // kernels launched by the current call (gcgt_stats.launches)
};

namespace {

constexpr int kBlock = 256;
#ifndef GCGT_EXPAND_MINB
#define GCGT_EXPAND_MINB 4  // resident expand blocks per SM the register budget is sized for (64 regs)
#endif
constexpr int kWarps = kBlock / 32;
// A vertex with more residual segments than this is not expanded by its own warp: its segments go to the
// level's hub queue and are spread over the whole grid (segment-level work stealing, the B200 analogue of the
// paper's Task Stealing + Residual Segmentation, §4.3 :884-930, §5.2 :1092-1136).

__device__ __forceinline__ uint32_t lane_id() { return threadIdx.x & 31; }
__device__ __forceinline__ uint32_t lanemask_lt() { uint32_t m; asm("mov.u32 %0, %%lanemask_lt;" : "=r"(m)); return m; }

// Kernel-constant view of the device CGR plus the per-level hub queue.
struct Ctx {
    const uint64_t* __restrict__ W;
    const uint64_t* __restrict__ offs;
    uint32_t min_len;
    uint32_t seg_bits;
    HubEntry* hubq;
    unsigned long long* hub_ctr;  // (entries << 32) | segments
    Stats* st;
    unsigned long long* cursor;   // work cursor over the frontier queue (reset per launch)
    HeavyEntry* heavyq;           // per-level heavy-vertex queue
    uint32_t* heavy_len;
    uint32_t heavy_itv;           // interval count above which a vertex is deferred to the heavy pass
    uint32_t heavy_res;           // unsegmented residual count above which a vertex is deferred
    uint32_t hub_segs;            // segment count above which a vertex's segments go to the hub queue
    uint32_t engine;              // 1 = state-machine kernel (sm_expand_kernel), 0 = phase kernel (expand_kernel)
    const uint32_t* dir;          // BFS direction gate: top-down kernels run only while *dir == 0 (nullptr: always)
    // interval checkpoints (vertices with more than ck_c intervals; sorted ids, per-vertex checkpoint ranges)
    uint32_t hv_n, ck_c;
    const uint32_t* __restrict__ hv_ids;
    const uint32_t* __restrict__ hv_ptr;
    const uint32_t* __restrict__ hv_wptr;  // per-word index (hv_index), words from hv_w0
    const uint32_t* __restrict__ hv_bits;
    uint64_t hv_w0;
    const uint64_t* __restrict__ hv_after;  // bit after the interval area
    const uint32_t* __restrict__ hv_rem;    // unsegmented records: residual count
    const uint64_t* __restrict__ ck_pos;
    const uint32_t* __restrict__ ck_prev;
    LongRange* lrq;
    unsigned long long* lr_ctr;
    uint32_t long_len, lr_chunk;
    // fused hub consumption (expand_kernel drains the level's hub segments / long ranges itself, no hub_kernel):
    // fuse_ctr[0] blocks done expanding, [1] long-range take cursor, [2] hub-segment take cursor, [3] epoch
    uint32_t fuse;
    uint32_t* fuse_ctr;
    uint32_t flatb;  // phase B as a lane-refill loop (1) or in static rounds of 32 tasks (0)
};

// Publication of hub / long-range entries: the data, a fence, then the launch's epoch (the readiness flag).
__device__ __forceinline__ void publish_hub(HubEntry* q, uint64_t idx, uint64_t base, uint32_t u, uint32_t off,
                                            uint32_t epoch) {
    HubEntry* e = q + idx;
    e->base = base;
    e->u = u;
    e->seg_off = off;
    __threadfence();
    *(volatile uint32_t*)&e->epoch = epoch;
}
__device__ __forceinline__ void publish_lr(LongRange* q, uint64_t idx, uint32_t u, uint32_t start, uint32_t len,
                                           uint32_t off, uint32_t epoch) {
    LongRange* e = q + idx;
    e->u = u;
    e->start = start;
    e->len = len;
    e->chunk_off = off;
    __threadfence();
    *(volatile uint32_t*)&e->epoch = epoch;
}
__device__ __forceinline__ uint32_t cur_epoch(const Ctx& c) {
    return c.fuse_ctr ? *(volatile const uint32_t*)(c.fuse_ctr + 3) : 0u;
}

__device__ __forceinline__ void add_stats(Stats* st, uint64_t v, uint64_t a, uint64_t b) {
    for (int o = 16; o; o >>= 1) {  // warp reduce (call with the full warp), one atomic per warp
        v += __shfl_xor_sync(0xffffffffu, v, o);
        a += __shfl_xor_sync(0xffffffffu, a, o);
        b += __shfl_xor_sync(0xffffffffu, b, o);
    }
    if (lane_id() == 0 && (v | a | b)) {
        if (v) atomicAdd(&st->vertices, (unsigned long long)v);
        if (a) atomicAdd(&st->arcs, (unsigned long long)a);
        if (b) atomicAdd(&st->bits, (unsigned long long)b);
    }
}

// ---- frontier sources ------------------------------------------------------------------------------------------------
// Queue of frontier words (BFS / BC): entry i is word q[i]; its bits come from qbits[i] (BC keeps them per level)
// or from the frontier bitmap F (BFS; the contraction rewrites F densely every level).
struct QueueFront {
    const uint32_t* __restrict__ q;
    const uint32_t* __restrict__ qlen_p;
    uint32_t* __restrict__ F;
    const uint32_t* __restrict__ qbits;
    __device__ __forceinline__ uint64_t size() const { return *qlen_p; }
    __device__ __forceinline__ void get(uint64_t i, uint32_t& w, uint32_t& bits) const {
        w = q[i];
        bits = qbits ? qbits[i] : F[w];
    }
};

// The level's heavy-vertex queue: one vertex per entry.
struct HeavyFront {
    const HeavyEntry* __restrict__ q;
    const uint32_t* __restrict__ len_p;
    __device__ __forceinline__ uint64_t size() const { return *len_p; }
    __device__ __forceinline__ void get(uint64_t i, uint32_t& w, uint32_t& bits) const {
        const uint32_t u = q[i].u;
        w = u >> 5;
        bits = 1u << (u & 31);
    }
};

// Frontier bits of the owned word range (partitioned BFS): entry i is word w_lo + i with its F bits restricted to
// the owned vertices [lo, hi).
struct BitsFront {
    const uint32_t* __restrict__ F;
    uint64_t lo, hi;
    __device__ __forceinline__ uint64_t size() const { return hi > lo ? ((hi + 31) >> 5) - (lo >> 5) : 0; }
    __device__ __forceinline__ void get(uint64_t i, uint32_t& w, uint32_t& bits) const {
        w = (uint32_t)((lo >> 5) + i);
        const uint64_t v0 = (uint64_t)w * 32;
        bits = F[w];
        if (v0 < lo) bits &= 0xffffffffu << (lo - v0);
        if (v0 + 32 > hi) bits &= (hi - v0 >= 32) ? 0xffffffffu : ((1u << (hi - v0)) - 1);
    }
};

// Every vertex of [lo, hi) (CC's hooking pass).
struct DenseFront {
    uint64_t lo, hi;
    __device__ __forceinline__ uint64_t size() const { return hi > lo ? ((hi + 31) >> 5) - (lo >> 5) : 0; }
    __device__ __forceinline__ void get(uint64_t i, uint32_t& w, uint32_t& bits) const {
        w = (uint32_t)((lo >> 5) + i);
        const uint64_t v0 = (uint64_t)w * 32;
        bits = 0xffffffffu;
        if (v0 < lo) bits &= 0xffffffffu << (lo - v0);
        if (v0 + 32 > hi) bits &= (hi - v0 >= 32) ? 0xffffffffu : ((1u << (hi - v0)) - 1);
    }
};

// ---- decode helpers ---------------------------------------------------------------------------------------------------
// One residual segment (FORMAT.md R17): count, first residual anchored at u, then gaps.  Returns the count.
// The segment's bits are staged in registers (RegStream) and the neighbour ids are handed to the filter four at a
// time (App::many), so their visited-bitmap probes are in flight together.
// Interval hand-off: short intervals go to the filter directly; long ones to the level's long-range queue.
template <class App>
__device__ __forceinline__ void range_or_defer(const Ctx& c, App& t, uint32_t u, uint32_t start, uint32_t len) {
    if (len <= c.long_len || !c.lr_ctr) {
        t.range(start, len);
        return;
    }
    const uint32_t nch = (len + c.lr_chunk - 1) / c.lr_chunk;
    const unsigned long long old = atomicAdd(c.lr_ctr, (1ull << 32) | (unsigned long long)nch);
    publish_lr(c.lrq, old >> 32, u, start, len, (uint32_t)(old & 0xffffffffu), cur_epoch(c));
}

// Per-codeword global-window reader (the unstaged alternative to RegStream; same interface).
struct WinStream {
    const uint64_t* __restrict__ W;
    uint64_t p;
    __device__ __forceinline__ void init(const uint64_t* __restrict__ w, uint64_t pos) { W = w; p = pos; }
    template <int K>
    __device__ __forceinline__ uint64_t next() { return decode<K>(W, p); }
};

// Sequential reader over BitBuf (the 32-bit refill bit buffer); same interface.
struct BufStream {
    const uint64_t* __restrict__ W;
    BitBuf bb;
    uint64_t p;  // only meaningful after sync()
    __device__ __forceinline__ void init(const uint64_t* __restrict__ w, uint64_t pos) {
        W = w;
        bb.init(w, pos);
        p = pos;
    }
    template <int K>
    __device__ __forceinline__ uint64_t next() {
        const uint64_t v = bb.template next<K>(W);
        p = bb.pos();
        return v;
    }
};

template <bool STAGED>
using Reader = typename std::conditional<STAGED, BufStream, WinStream>::type;

template <int K, bool STAGED, class T>
__device__ __forceinline__ uint32_t decode_segment(const uint64_t* __restrict__ W, uint64_t q, uint32_t u, T& t) {
    Reader<STAGED> rs;
    rs.init(W, q);
    const uint32_t cnt = (uint32_t)(rs.template next<K>() - 1);
    int64_t cur = 0;
    for (uint32_t done = 0; done < cnt; done += 4) {
        uint32_t v[4];
        const uint32_t nb = min(4u, cnt - done);
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            if (k < nb) {
                const uint64_t c = rs.template next<K>();
                cur = (done + k == 0) ? unmap_first(u, c) : cur + (int64_t)c;
                v[k] = (uint32_t)cur;
            }
        }
        t.many(v, nb);
    }
    return cnt;
}

// ---- the expansion engine -----------------------------------------------------------------------------------------
// Work distribution: a persistent grid (one wave, sized by the occupancy calculator) whose warps grab `wpb` queue
// words at a time from an atomic cursor (dynamic load balancing; no tail of idle SMs).  For each batch:
// Phase A (lane per frontier vertex): App::vertex, the record header and the interval area (decoded serially, each
//   interval handed over as a word-range claim), then segNum.  A vertex whose interval area (or unsegmented list)
//   is long is deferred as "heavy".
// Phase B (segmented format): the batch's segments are flattened with a warp scan and decoded one segment per
//   lane (segments are self-contained, R17), so lane work is bounded by 2 segBits bits regardless of degree.
//   Vertices with more than kHubSegs segments go to the hub queue (hub_kernel, whole grid).
// Heavy vertices (long interval area, or long unsegmented list) go to the level's heavy queue, which a second
//   pass of the same kernel (DEFER = false) drains one lane per heavy vertex over the whole grid, so a long
//   record never stalls a batch.  (A whole-warp Alg. 4 decode of the long record was measured slower on B200:
//   each window step is a ~1.5k-cycle dependent chain for ~5 codewords vs ~60 cycles per codeword serially;
//   DESIGN.md §6.)

struct WarpSmem {
    uint32_t w[32], b[32], pre[33];
    uint32_t u[32], spre[33];
    uint64_t base[32];
    uint32_t ckb[32], nck[32], itv[32];  // interval-chunk tasks of long interval areas (checkpoint table)
    uint32_t take;                       // phase-B work cursor (lane-refill loop)
};

// DEFER = true: the level's frontier pass (heavy vertices are queued); false: the heavy pass over that queue
// (same engine, one lane per heavy vertex, nothing deferred, App::vertex and vertex stats already done).
template <int K, bool SEG, class App, class Front, bool DEFER, bool STAGED>
__device__ __forceinline__ void expand_phase(const Ctx& c, const Front& fr, const App& app, uint32_t wpb,
                                             WarpSmem* smem, uint64_t& nv, uint64_t& na, uint64_t& nb) {
    const uint32_t wid = threadIdx.x >> 5, lane = lane_id();
    WarpSmem& sm = smem[wid];
    if (c.dir && *c.dir) return;  // this level runs bottom-up
    const uint64_t qlen = fr.size();
    if (wpb == 0) {  // sized on the device (host did not wait for the queue length): ~4 batches per resident warp
        const uint64_t b = qlen / ((uint64_t)gridDim.x * kWarps * 4);
        wpb = b < 1 ? 1 : (b > 8 ? 8 : (uint32_t)b);
    }
    // Every warp's first batch is static (its global warp index), so a small frontier costs no cursor atomics; later
    // batches come from the atomic cursor, numbered after the static ones and fetched one batch ahead.
    const uint64_t nstatic = (uint64_t)gridDim.x * kWarps * wpb;
    unsigned long long next = ((uint64_t)blockIdx.x * kWarps + wid) * wpb;
    for (;;) {
        const uint64_t base = __shfl_sync(0xffffffffu, next, 0);
        if (base >= qlen) break;
        if (lane == 0) next = nstatic + atomicAdd(c.cursor, (unsigned long long)wpb);
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
            // ---- phase A
            const uint32_t j = t0 + lane;
            uint32_t nseg = 0, u = 0, ckb = 0, nck = 0, itv_all = 0;
            uint64_t segbase = 0;
            if (j < total) {
                uint32_t lo = 0, hi = 31;  // owner lane: largest o with pre[o] <= j
                while (lo < hi) {
                    const uint32_t mid = (lo + hi + 1) >> 1;
                    if (sm.pre[mid] <= j) lo = mid; else hi = mid - 1;
                }
                u = sm.w[lo] * 32 + __fns(sm.b[lo], 0, (int)(j - sm.pre[lo]) + 1);
                uint64_t p = ldg64(c.offs + u);
                App t = app;
                t.begin(u);
                if (DEFER) {
                    nb += ldg64(c.offs + u + 1) - p;
                    nv++;
                    t.vertex(u);
                }
                Reader<STAGED> rs;
                rs.init(c.W, p);
                uint64_t deg = 0;
                if (!SEG) deg = rs.template next<K>() - 1;
                const uint64_t itv = rs.template next<K>() - 1;
                p = rs.p;
                if (DEFER && (itv > c.heavy_itv || (!SEG && deg > c.heavy_res))) {  // heavy: deferred to the heavy pass
                    cg::coalesced_group grp = cg::coalesced_threads();
                    uint32_t slot = 0;
                    if (grp.thread_rank() == 0) slot = atomicAdd(c.heavy_len, grp.size());
                    slot = grp.shfl(slot, 0) + grp.thread_rank();
                    c.heavyq[slot] = HeavyEntry{p, u, (uint32_t)itv, deg};
                } else {
                    int64_t prev_end = 0;
                    uint64_t in_itv = 0, nres_ck = 0;
                    uint64_t itv_here = itv;
                    bool ck = false;
                    uint64_t after = 0;
                    if (c.hv_n && itv > c.ck_c) {  // long interval area: chunks beyond the first go grid-wide
                        const uint64_t wl = (u >> 5) - c.hv_w0;
                        const uint32_t lo = c.hv_wptr[wl] + __popc(c.hv_bits[wl] & ((1u << (u & 31)) - 1));
                        ckb = c.hv_ptr[lo];  // chunks 1.. become phase-B tasks of this batch
                        nck = c.hv_ptr[lo + 1] - ckb;
                        itv_all = (uint32_t)itv;
                        itv_here = c.ck_c;
                        after = c.hv_after[lo];
                        if (!SEG) nres_ck = c.hv_rem[lo];
                        ck = true;
                    }
                    for (uint64_t i = 0; i < itv_here; i++) {
                        const uint64_t g = rs.template next<K>();
                        const uint64_t len = rs.template next<K>() - 1 + c.min_len;
                        const int64_t start = i == 0 ? unmap_first(u, g) : prev_end + (int64_t)g;
                        range_or_defer(c, t, u, (uint32_t)start, (uint32_t)len);
                        prev_end = start + (int64_t)len - 1;
                        in_itv += len;
                    }
                    na += in_itv;
                    if (ck) rs.init(c.W, after);
                    if (!SEG) {
                        const uint64_t nres = ck ? nres_ck : deg - in_itv;
                        int64_t cur = 0;
                        for (uint64_t i = 0; i < nres; i++) {
                            const uint64_t cd = rs.template next<K>();
                            cur = i == 0 ? unmap_first(u, cd) : cur + (int64_t)cd;
                            t.one((uint32_t)cur);
                        }
                        na += nres;
                    } else {
                        nseg = (uint32_t)(rs.template next<K>() - 1);
                        segbase = rs.p;
                        if (nseg > c.hub_segs || (!DEFER && nseg)) {  // hub: hand the segments to the whole grid
                            const unsigned long long old =
                                atomicAdd(c.hub_ctr, (1ull << 32) | (unsigned long long)nseg);
                            publish_hub(c.hubq, old >> 32, segbase, u, (uint32_t)(old & 0xffffffffu), cur_epoch(c));
                            nseg = 0;
                        }
                    }
                    t.end();
                }
            }
            if (SEG || c.hv_n) {
                // ---- phase B: flatten the batch's tasks (interval chunks, then residual segments), one per lane
                uint32_t sincl = nck + nseg;
                for (int o = 1; o < 32; o <<= 1) {
                    const uint32_t tt = __shfl_up_sync(0xffffffffu, sincl, o);
                    if (lane >= (uint32_t)o) sincl += tt;
                }
                sm.u[lane] = u;
                sm.base[lane] = segbase;
                sm.ckb[lane] = ckb;
                sm.nck[lane] = nck;
                sm.itv[lane] = itv_all;
                sm.spre[lane + 1] = sincl;
                if (lane == 0) sm.spre[0] = 0;
                if (lane == 0) sm.take = 32;
                __syncwarp();
                const uint32_t stotal = sm.spre[32];
                if (c.flatb) {
                    // lane-refill loop: a lane that finishes its task takes the next one at once (warp-local work
                    // cursor), so a round no longer waits for its longest segment; segments are decoded four
                    // codewords per iteration (one batched probe per four ids)
                    uint32_t sj = lane, rem = 0, su = 0;
                    uint64_t sp = 0;
                    int64_t scur = 0;
                    bool sfirst = false, open = false;
                    App t = app;
                    for (;;) {
                        if (rem == 0) {
                            if (open) {
                                t.end();
                                open = false;
                            }
                            if (sj >= stotal) break;
                            uint32_t lo = 0, hi = 31;
                            while (lo < hi) {
                                const uint32_t mid = (lo + hi + 1) >> 1;
                                if (sm.spre[mid] <= sj) lo = mid; else hi = mid - 1;
                            }
                            su = sm.u[lo];
                            const uint32_t idx = sj - sm.spre[lo], snck = sm.nck[lo];
                            t = app;
                            t.begin(su);
                            open = true;
                            if (idx < snck) {  // interval chunk idx+1 of su, processed whole
                                const uint32_t k = sm.ckb[lo] + idx;
                                const uint32_t left = sm.itv[lo] - (idx + 1) * c.ck_c;
                                const uint32_t cnt = left < c.ck_c ? left : c.ck_c;
                                uint64_t p = c.ck_pos[k];
                                uint32_t cur = c.ck_prev[k];
                                for (uint32_t i = 0; i < cnt; i++) {
                                    const uint32_t g = (uint32_t)decode<K>(c.W, p);
                                    const uint32_t len = (uint32_t)(decode<K>(c.W, p) - 1) + c.min_len;
                                    range_or_defer(c, t, su, cur + g, len);
                                    cur += g + len - 1;
                                    na += len;
                                }
                            } else {
                                sp = sm.base[lo] + (uint64_t)(idx - snck) * c.seg_bits;
                                rem = (uint32_t)(decode<K>(c.W, sp) - 1);
                                na += rem;
                                sfirst = true;
                            }
                            sj = atomicAdd(&sm.take, 1u);
                            continue;
                        }
                        uint32_t v[4];
                        const uint32_t nb = min(4u, rem);
#pragma unroll
                        for (uint32_t k = 0; k < 4; k++) {
                            if (k < nb) {
                                const uint64_t cw = decode<K>(c.W, sp);
                                scur = sfirst ? unmap_first(su, cw) : scur + (int64_t)cw;
                                sfirst = false;
                                v[k] = (uint32_t)scur;
                            }
                        }
                        t.many(v, nb);
                        rem -= nb;
                    }
                } else
                for (uint32_t k0 = 0; k0 < stotal; k0 += 32) {
                    const uint32_t sj = k0 + lane;
                    if (sj < stotal) {
                        uint32_t lo = 0, hi = 31;
                        while (lo < hi) {
                            const uint32_t mid = (lo + hi + 1) >> 1;
                            if (sm.spre[mid] <= sj) lo = mid; else hi = mid - 1;
                        }
                        const uint32_t su = sm.u[lo], idx = sj - sm.spre[lo], snck = sm.nck[lo];
                        App t = app;
                        t.begin(su);
                        if (idx < snck) {  // interval chunk idx+1 of su: up to ck_c intervals from a checkpoint
                            const uint32_t k = sm.ckb[lo] + idx;
                            const uint32_t left = sm.itv[lo] - (idx + 1) * c.ck_c;
                            const uint32_t cnt = left < c.ck_c ? left : c.ck_c;
                            uint64_t p = c.ck_pos[k];
                            uint32_t cur = c.ck_prev[k];
                            for (uint32_t i = 0; i < cnt; i++) {
                                const uint32_t g = (uint32_t)decode<K>(c.W, p);
                                const uint32_t len = (uint32_t)(decode<K>(c.W, p) - 1) + c.min_len;
                                range_or_defer(c, t, su, cur + g, len);
                                cur += g + len - 1;
                                na += len;
                            }
                        } else {
                            na += decode_segment<K, STAGED>(c.W, sm.base[lo] + (uint64_t)(idx - snck) * c.seg_bits,
                                                            su, t);
                        }
                        t.end();
                    }
                }
            }
            __syncwarp();
        }
        __syncwarp();
    }
}

// Fused hub consumption (Ctx::fuse): a block that has finished its share of the frontier drains the level's hub
// segments and long-range chunks while other blocks are still expanding (and publishing more), instead of a separate
// hub_kernel launch after the whole expansion.  Warps claim 32 items at a time from a take cursor; an item whose
// entry is not yet published is waited for; the queues are final once every block has finished expanding (the
// grid is one co-resident wave, so waiting cannot deadlock).  Entry reads bypass L1 (volatile): they are written
// by other SMs during this launch.
__device__ __forceinline__ uint32_t entry_off(const volatile HubEntry* e) { return e->seg_off; }
__device__ __forceinline__ uint32_t entry_off(const volatile LongRange* e) { return e->chunk_off; }
template <class E>
__device__ __forceinline__ uint32_t find_entry(const E* q, uint32_t ne, uint32_t j, uint32_t epoch) {
    uint32_t lo = 0, hi = ne - 1;  // largest entry whose offset is <= j (entries are ordered by offset)
    while (lo < hi) {
        const uint32_t mid = (lo + hi + 1) >> 1;
        const volatile E* e = q + mid;
        while (e->epoch != epoch) __nanosleep(32);
        if (entry_off(e) <= j) lo = mid; else hi = mid - 1;
    }
    const volatile E* e = q + lo;
    while (e->epoch != epoch) __nanosleep(32);
    __threadfence();
    return lo;
}

__device__ __forceinline__ uint32_t ld_acquire(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ unsigned long long ld_acquire(const unsigned long long* p) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}

template <int K, bool STAGED, class App>
__device__ __forceinline__ void hub_consume(const Ctx& c, const App& app, uint32_t epoch, uint64_t& na) {
    const uint32_t lane = lane_id();
    uint32_t* fc = c.fuse_ctr;
    for (;;) {
        const uint32_t done = ld_acquire(fc);
        const unsigned long long lc = ld_acquire(c.lr_ctr);
        const unsigned long long hc = ld_acquire(c.hub_ctr);
        const bool final = done == gridDim.x;
        const uint32_t lt = ld_acquire(fc + 1), ht = ld_acquire(fc + 2);
        int qsel;
        if (lt < (uint32_t)lc) qsel = 0;
        else if (ht < (uint32_t)hc) qsel = 1;
        else if (final) return;
        else {
            __nanosleep(500);
            continue;
        }
        uint32_t j0 = 0;
        if (lane == 0) j0 = atomicAdd(fc + 1 + qsel, 32u);
        j0 = __shfl_sync(0xffffffffu, j0, 0);
        const uint32_t j = j0 + lane;
        bool pending = true;
        for (;;) {
            const uint32_t dn = ld_acquire(fc);
            const unsigned long long cv = ld_acquire(qsel == 0 ? c.lr_ctr : c.hub_ctr);
            const uint32_t S = (uint32_t)cv, ne = (uint32_t)(cv >> 32);
            if (pending && j < S) {
                pending = false;
                App t = app;
                if (qsel == 0) {
                    const uint32_t k = find_entry(c.lrq, ne, j, epoch);
                    const volatile LongRange* e = c.lrq + k;
                    const uint32_t eu = e->u, es = e->start, el = e->len, eo = e->chunk_off;
                    const uint32_t off = (j - eo) * c.lr_chunk;
                    t.begin(eu);
                    t.range(es + off, min(c.lr_chunk, el - off));
                    t.end();
                } else {
                    const uint32_t k = find_entry(c.hubq, ne, j, epoch);
                    const volatile HubEntry* e = c.hubq + k;
                    const uint64_t eb = e->base;
                    const uint32_t eu = e->u, eo = e->seg_off;
                    t.begin(eu);
                    na += decode_segment<K, STAGED>(c.W, eb + (uint64_t)(j - eo) * c.seg_bits, eu, t);
                    t.end();
                }
            }
            const bool fin = dn == gridDim.x;
            if (__all_sync(0xffffffffu, !pending || (fin && j >= S))) break;
            __nanosleep(200);
        }
    }
}

template <int K, bool SEG, class App, class Front, bool DEFER, bool STAGED>
__global__ void __launch_bounds__(kBlock, GCGT_EXPAND_MINB) expand_kernel(Ctx c, Front fr, App app, uint32_t wpb) {
    __shared__ WarpSmem smem[kWarps];
    if (c.dir && *c.dir) return;  // this BFS level runs bottom-up: no work, cursor untouched
    uint64_t nv = 0, na = 0, nb = 0;
    const bool fuse = DEFER && c.fuse;
    const uint32_t epoch = fuse ? cur_epoch(c) : 0u;
    expand_phase<K, SEG, App, Front, DEFER, STAGED>(c, fr, app, wpb, smem, nv, na, nb);
    if (fuse) {
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            atomicAdd(c.fuse_ctr, 1u);
        }
        if ((threadIdx.x >> 5) < c.fuse) hub_consume<K, STAGED>(c, app, epoch, na);  // c.fuse consumer warps per block
    }
    add_stats(c.st, nv, na, nb);
    // the last block out resets the work cursor (and the fused-hub counters, advancing the epoch) for the next launch
    __syncthreads();
    if (threadIdx.x == 0) {
        if (atomicAdd(c.cursor + 1, 1ull) == gridDim.x - 1) {
            c.cursor[0] = 0;
            c.cursor[1] = 0;
            if (fuse) {
                c.fuse_ctr[0] = 0;
                c.fuse_ctr[1] = 0;
                c.fuse_ctr[2] = 0;
                c.fuse_ctr[3] = epoch + 1;
            }
        }
    }
}

// ---- the state-machine expansion kernel (default) ---------------------------------------------------------------
// Every lane runs a small state machine over "tasks": a vertex task decodes the record header and the interval
// area (each interval handed over as a range claim) and queues the vertex's residual segments; a segment task
// decodes one residual segment (FORMAT.md R17).  Each loop iteration every busy lane decodes exactly ONE codeword
// (BitBuf) and acts on it, so the warp's lanes stay busy regardless of how skewed the records are; lanes that
// finish take the next task at a warp-uniform refill point: first segments from the warp's ring (64 entries in
// shared memory), then vertices of the current frontier batch, fetching a new batch from the global work cursor
// when the batch is used up.  This is the paper's Task Stealing (Alg. 3, §4.3 :884-930) and Residual Segmentation
// (§5.2) recast as a warp-level scheduler: idle lanes steal whole segments instead of decoded neighbours.
// Vertices with more than hub_segs segments (or overflowing the ring) go to the grid-wide hub queue.
constexpr uint32_t kRing = 64;
constexpr uint32_t kList = 256;  // 8 queue words x 32 vertices

struct SmWarp {
    uint32_t list[kList];
    uint32_t ring_u[kRing];
    uint64_t ring_p[kRing];
    uint32_t head, tail;
};

enum : uint32_t { ST_DONE = 0, ST_DEG, ST_ITVN, ST_GAP, ST_LEN, ST_SEGN, ST_RES, ST_SCNT, ST_SFIRST, ST_SGAP };

template <int K, bool SEG, class App, class Front>
__global__ void __launch_bounds__(kBlock, 4) sm_expand_kernel(Ctx c, Front fr, App app, uint32_t wpb) {
    __shared__ SmWarp smem[kWarps];
    const uint32_t wid = threadIdx.x >> 5, lane = lane_id(), lt = lanemask_lt();
    SmWarp& sm = smem[wid];
    const uint64_t qlen = (c.dir && *c.dir) ? 0 : fr.size();
    if (wpb == 0) {
        const uint64_t b = qlen / ((uint64_t)gridDim.x * kWarps * 4);
        wpb = b < 1 ? 1 : (b > 8 ? 8 : (uint32_t)b);
    }
    if (wpb > kList / 32) wpb = kList / 32;
    if (lane == 0) sm.head = sm.tail = 0;
    uint32_t list_n = 0, list_pos = 0;  // warp-uniform
    bool cursor_done = false;
    unsigned long long next = 0;
    if (lane == 0) next = atomicAdd(c.cursor, (unsigned long long)wpb);
    // per-lane task state
    uint32_t state = ST_DONE, u = 0, i = 0, cnt = 0, start = 0, cur = 0, push_n = 0;
    uint64_t push_base = 0, rem = 0;
    BitBuf bb{0, 0, 0};
    App t = app;
    uint64_t nv = 0, na = 0, nb = 0;
    __syncwarp();
    for (;;) {
        // ---- queue the segments produced by the last step (warp scan over the pushes)
        const uint32_t pmask = __ballot_sync(0xffffffffu, push_n != 0);
        if (pmask) {
            uint32_t incl = push_n;
            for (int o = 1; o < 32; o <<= 1) {
                const uint32_t tt = __shfl_up_sync(0xffffffffu, incl, o);
                if (lane >= (uint32_t)o) incl += tt;
            }
            const uint32_t head = sm.head, tail = sm.tail, space = kRing - (tail - head);
            if (push_n) {
                const uint32_t off = incl - push_n;
                if (incl <= space) {
                    for (uint32_t k = 0; k < push_n; k++) {
                        const uint32_t slot = (tail + off + k) % kRing;
                        sm.ring_u[slot] = u;
                        sm.ring_p[slot] = push_base + (uint64_t)k * c.seg_bits;
                    }
                } else {  // ring full: the grid-wide hub queue takes them
                    const unsigned long long old = atomicAdd(c.hub_ctr, (1ull << 32) | (unsigned long long)push_n);
                    publish_hub(c.hubq, old >> 32, push_base, u, (uint32_t)(old & 0xffffffffu), cur_epoch(c));
                }
                push_n = 0;
            }
            __syncwarp();
            // pushes are stored in lane order while they fit, so the stored ones are a prefix of the pushers
            const uint32_t stored = __reduce_max_sync(0xffffffffu, (incl <= space && (pmask >> lane) & 1u) ? incl : 0u);
            if (lane == 0) sm.tail = tail + stored;
            __syncwarp();
        }
        // ---- refill idle lanes (warp-uniform)
        uint32_t idle = __ballot_sync(0xffffffffu, state == ST_DONE);
        if (idle) {
            const uint32_t head = sm.head, avail = sm.tail - head;
            if (avail) {
                const uint32_t r = __popc(idle & lt), take = min(avail, (uint32_t)__popc(idle));
                if (state == ST_DONE && r < take) {
                    const uint32_t slot = (head + r) % kRing;
                    u = sm.ring_u[slot];
                    bb.init(c.W, sm.ring_p[slot]);
                    t = app;
                    t.begin(u);
                    state = ST_SCNT;
                }
                __syncwarp();
                if (lane == 0) sm.head = head + take;
                __syncwarp();
                idle = __ballot_sync(0xffffffffu, state == ST_DONE);
            }
            while (idle) {
                if (list_pos >= list_n) {
                    if (cursor_done) break;
                    const uint64_t base = __shfl_sync(0xffffffffu, next, 0);
                    if (base >= qlen) {
                        cursor_done = true;
                        break;
                    }
                    if (lane == 0) next = atomicAdd(c.cursor, (unsigned long long)wpb);
                    uint32_t w = 0, bits = 0;
                    if (lane < wpb && base + lane < qlen) fr.get(base + lane, w, bits);
                    uint32_t incl = __popc(bits);
                    for (int o = 1; o < 32; o <<= 1) {
                        const uint32_t tt = __shfl_up_sync(0xffffffffu, incl, o);
                        if (lane >= (uint32_t)o) incl += tt;
                    }
                    uint32_t pos = incl - __popc(bits);
                    for (uint32_t bm = bits; bm; bm &= bm - 1) sm.list[pos++] = w * 32 + (__ffs(bm) - 1);
                    list_n = __shfl_sync(0xffffffffu, incl, 31);
                    list_pos = 0;
                    __syncwarp();
                    continue;
                }
                const uint32_t r = __popc(idle & lt), take = min(list_n - list_pos, (uint32_t)__popc(idle));
                if (state == ST_DONE && r < take) {
                    u = sm.list[list_pos + r];
                    const uint64_t p = ldg64(c.offs + u);
                    nb += ldg64(c.offs + u + 1) - p;
                    nv++;
                    t = app;
                    t.begin(u);
                    t.vertex(u);
                    bb.init(c.W, p);
                    state = SEG ? ST_ITVN : ST_DEG;
                }
                list_pos += take;
                idle = __ballot_sync(0xffffffffu, state == ST_DONE);
            }
            if (idle == 0xffffffffu) {
                if (cursor_done && list_pos >= list_n && sm.head == sm.tail) break;
                continue;  // (cannot happen with work pending; defensive)
            }
        }
        // ---- one step: every busy lane decodes one codeword and acts on it
        if (state != ST_DONE) {
            const uint64_t v = bb.template next<K>(c.W);
            bool itv_done = false;
            switch (state) {
                case ST_DEG:
                    rem = v - 1;
                    state = ST_ITVN;
                    break;
                case ST_ITVN:
                    cnt = (uint32_t)(v - 1);
                    i = 0;
                    if (cnt) state = ST_GAP;
                    else itv_done = true;
                    break;
                case ST_GAP:
                    start = i == 0 ? (uint32_t)unmap_first(u, v) : cur + (uint32_t)v;
                    state = ST_LEN;
                    break;
                case ST_LEN: {
                    const uint32_t len = (uint32_t)(v - 1) + c.min_len;
                    t.range(start, len);
                    na += len;
                    if (!SEG) rem -= len;
                    cur = start + len - 1;
                    if (++i < cnt) state = ST_GAP;
                    else itv_done = true;
                    break;
                }
                case ST_SEGN: {
                    const uint32_t nseg = (uint32_t)(v - 1);
                    t.end();
                    state = ST_DONE;
                    if (nseg > c.hub_segs) {
                        const unsigned long long old = atomicAdd(c.hub_ctr, (1ull << 32) | (unsigned long long)nseg);
                        publish_hub(c.hubq, old >> 32, bb.pos(), u, (uint32_t)(old & 0xffffffffu), cur_epoch(c));
                    } else if (nseg) {
                        push_n = nseg;
                        push_base = bb.pos();
                    }
                    break;
                }
                case ST_RES:
                    cur = i == 0 ? (uint32_t)unmap_first(u, v) : cur + (uint32_t)v;
                    t.one(cur);
                    na++;
                    if (++i == rem) {
                        t.end();
                        state = ST_DONE;
                    }
                    break;
                case ST_SCNT:
                    cnt = (uint32_t)(v - 1);
                    i = 0;
                    state = ST_SFIRST;
                    break;
                case ST_SFIRST:
                    cur = (uint32_t)unmap_first(u, v);
                    t.one(cur);
                    na++;
                    if (++i == cnt) {
                        t.end();
                        state = ST_DONE;
                    } else {
                        state = ST_SGAP;
                    }
                    break;
                case ST_SGAP:
                    cur += (uint32_t)v;
                    t.one(cur);
                    na++;
                    if (++i == cnt) {
                        t.end();
                        state = ST_DONE;
                    }
                    break;
            }
            if (itv_done) {
                if (SEG) {
                    state = ST_SEGN;
                } else if (rem) {
                    state = ST_RES;
                    i = 0;
                } else {
                    t.end();
                    state = ST_DONE;
                }
            }
        }
        __syncwarp();
    }
    add_stats(c.st, nv, na, nb);
    if (lane == 0) {
        const unsigned long long nw = (unsigned long long)gridDim.x * kWarps;
        if (atomicAdd(c.cursor + 1, 1ull) == nw - 1) {
            c.cursor[0] = 0;
            c.cursor[1] = 0;
        }
    }
}

// Entry of flattened item j in a queue ordered by offset (HubEntry::seg_off / LongRange::chunk_off), found by the
// whole warp at once: a 32-ary search for the warp's first item jb (ballot over 32 probes per round, ~log32(ne)
// dependent loads instead of ~log2(ne)), then each lane walks forward to its own item (entries hold >= 5 items).
__device__ __forceinline__ uint32_t item_off(const HubEntry* e) { return e->seg_off; }
__device__ __forceinline__ uint32_t item_off(const LongRange* e) { return e->chunk_off; }
template <class E>
__device__ __forceinline__ uint32_t warp_find_item(const E* __restrict__ q, uint32_t ne, uint32_t jb, uint32_t j) {
    const uint32_t lane = lane_id();
    uint32_t lo = 0, hi = ne;  // invariant: off[lo] <= jb, and off[hi] > jb if hi < ne
    while (hi - lo > 1) {
        const uint32_t span = hi - lo;
        const uint32_t pos = span <= 32 ? lo + lane : lo + (uint32_t)(((uint64_t)span * lane) >> 5);
        const bool le = (span > 32 || lane < span) && item_off(q + pos) <= jb;
        const uint32_t L = 31 - __clz(__ballot_sync(0xffffffffu, le));
        if (span <= 32) {
            lo += L;
            break;
        }
        const uint32_t nlo = lo + (uint32_t)(((uint64_t)span * L) >> 5);
        hi = L == 31 ? hi : lo + (uint32_t)(((uint64_t)span * (L + 1)) >> 5);
        lo = nlo;
    }
    uint32_t e = lo;
    while (e + 1 < ne && item_off(q + e + 1) <= j) e++;
    return e;
}

// Hub segments of the level, flattened over the whole grid (one segment per thread at a time).
template <int K, bool STAGED, class App>
__device__ __forceinline__ void hub_phase(const Ctx& c, const App& app, uint64_t& na) {
    const uint32_t lane = lane_id();
    const uint64_t gw0 = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) & ~31ull;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    if (c.lr_ctr) {  // long intervals: one lr_chunk-id piece per thread
        const unsigned long long lc = *(volatile unsigned long long*)c.lr_ctr;
        const uint32_t ne = (uint32_t)(lc >> 32), nchunks = (uint32_t)(lc & 0xffffffffu);
        for (uint64_t jb = gw0; jb < nchunks; jb += stride) {
            const uint32_t j = (uint32_t)jb + lane;
            const uint32_t k = warp_find_item(c.lrq, ne, (uint32_t)jb, min(j, nchunks - 1));
            if (j < nchunks) {
                const LongRange e = c.lrq[k];
                const uint32_t off = (j - e.chunk_off) * c.lr_chunk;
                App t = app;
                t.begin(e.u);
                t.range(e.start + off, min(c.lr_chunk, e.len - off));
                t.end();
            }
        }
    }
    const unsigned long long hc = *(volatile unsigned long long*)c.hub_ctr;
    const uint32_t nh = (uint32_t)(hc >> 32), S = (uint32_t)(hc & 0xffffffffu);
    for (uint64_t jb = gw0; jb < S; jb += stride) {
        const uint32_t j = (uint32_t)jb + lane;
        const uint32_t k = warp_find_item(c.hubq, nh, (uint32_t)jb, min(j, S - 1));
        if (j < S) {
            const HubEntry e = c.hubq[k];
            App t = app;
            t.begin(e.u);
            na += decode_segment<K, STAGED>(c.W, e.base + (j - e.seg_off) * (uint64_t)c.seg_bits, e.u, t);
            t.end();
        }
    }
}

template <int K, bool STAGED, class App>
__global__ void __launch_bounds__(kBlock) hub_kernel(Ctx c, App app) {
    if (*(volatile unsigned long long*)c.hub_ctr == 0 && (!c.lr_ctr || *(volatile unsigned long long*)c.lr_ctr == 0))
        return;  // no hub segments / long intervals this level
    uint64_t na = 0;
    hub_phase<K, STAGED>(c, app, na);
    add_stats(c.st, 0, na, 0);
}

// ---- applications (filters, Fig. 7) -------------------------------------------------------------------------------
// BFS (Fig. 7(b)).  V (visited, levels <= d) is immutable during a level, so it is read through the read-only path;
// a new vertex is claimed with a fire-and-forget atomicOr on the next-frontier bitmap N (no returned value on the
// critical path).  An interval is claimed 32 ids per atomic.
struct BfsApp {
    const uint32_t* __restrict__ V;
    uint32_t* __restrict__ N;
    int32_t* __restrict__ levels;
    int32_t level;
    uint32_t nfilter = 0;  // 1: skip the atomic when a (possibly stale) L1 read of N already shows the bits set
    __device__ __forceinline__ void begin(uint32_t) {}
    __device__ __forceinline__ void end() {}
    __device__ __forceinline__ void vertex(uint32_t) {}  // levels are written when a vertex is discovered
    // N is written concurrently: a plain (L1-cached, possibly stale) read can only under-report set bits, so
    // filtering on it never drops a claim; it only saves L2 atomics on vertices already claimed this level
    __device__ __forceinline__ static uint32_t ld_n(const uint32_t* p) {
        uint32_t v;
        asm volatile("ld.global.ca.u32 %0, [%1];" : "=r"(v) : "l"(p));
        return v;
    }
    __device__ __forceinline__ void claim(uint32_t w, uint32_t mask) {
        uint32_t cand = mask & ~__ldg(V + w);
        if (cand && nfilter) cand &= ~ld_n(N + w);
        if (cand) atomicOr(N + w, cand);
    }
    __device__ __forceinline__ void one(uint32_t v) { claim(v >> 5, 1u << (v & 31)); }
    // up to four ids: the four visited-bitmap probes are issued before any is consumed
    __device__ __forceinline__ void many(const uint32_t (&v)[4], uint32_t n) {
        uint32_t m[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) m[k] = k < n ? __ldg(V + (v[k] >> 5)) : 0xffffffffu;
        if (nfilter) {
#pragma unroll
            for (uint32_t k = 0; k < 4; k++)
                if (k < n && !(m[k] & (1u << (v[k] & 31)))) m[k] |= ld_n(N + (v[k] >> 5));
        }
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            const uint32_t bit = 1u << (v[k] & 31);
            if (k < n && !(m[k] & bit)) atomicOr(N + (v[k] >> 5), bit);
        }
    }
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        const uint32_t e = s + len;
        while (s < e) {
            const uint32_t b0 = s & 31, nb = min(32u - b0, e - s);
            claim(s >> 5, (nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0);
            s += nb;
        }
    }
};

// generic many() for filters without a batched form
#define GCGT_MANY_BY_ONE                                                         \
    __device__ __forceinline__ void many(const uint32_t (&v)[4], uint32_t n) {  \
        for (uint32_t k = 0; k < n; k++) one(v[k]);                              \
    }

// BC forward (Fig. 7(d), Brandes [9]): an arc u->v with v not in V (levels <= d) has level(v) = d+1, so
// sigma(v) += sigma(u); N collects level d+1.
struct BcFwdApp {
    const uint32_t* __restrict__ V;
    uint32_t* __restrict__ N;
    int32_t* __restrict__ levels;
    double* __restrict__ sigma;
    int32_t level;
    double su;
    __device__ __forceinline__ void begin(uint32_t u) { su = sigma[u]; }
    __device__ __forceinline__ void end() {}
    __device__ __forceinline__ void vertex(uint32_t u) { levels[u] = level; }
    __device__ __forceinline__ void claim(uint32_t w, uint32_t mask) {
        const uint32_t cand = mask & ~__ldg(V + w);
        if (!cand) return;
        atomicOr(N + w, cand);
        uint32_t cb = cand;
        while (cb) {
            const int b = __ffs(cb) - 1;
            cb &= cb - 1;
            atomicAdd(sigma + (uint64_t)w * 32 + b, su);
        }
    }
    __device__ __forceinline__ void one(uint32_t v) { claim(v >> 5, 1u << (v & 31)); }
    GCGT_MANY_BY_ONE
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        const uint32_t e = s + len;
        while (s < e) {
            const uint32_t b0 = s & 31, nb = min(32u - b0, e - s);
            claim(s >> 5, (nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0);
            s += nb;
        }
    }
};

// BC backward: delta(u) = sum_{w in out(u), d(w) = d(u)+1} sigma(u)/sigma(w) (1 + delta(w))  (Fig. 7(d)).
// A vertex's arcs are split over tasks (interval area + segments), so each task adds its partial sum to delta(u)
// and bc(u) (u != source); delta is zeroed per source.  Zero partials are skipped, so exact zeros stay exact.
struct BcBwdApp {
    const int32_t* __restrict__ levels;
    const double* __restrict__ sigma;
    double* __restrict__ delta;
    double* __restrict__ bc;
    int32_t next;
    uint32_t source;
    uint32_t u;
    double sv, acc;
    __device__ __forceinline__ void begin(uint32_t uu) { u = uu; sv = sigma[uu]; acc = 0.0; }
    __device__ __forceinline__ void vertex(uint32_t) {}
    __device__ __forceinline__ void one(uint32_t w) {
        if (levels[w] == next) acc += sv / sigma[w] * (1.0 + delta[w]);
    }
    GCGT_MANY_BY_ONE
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for (uint32_t t = 0; t < len; t++) one(s + t);
    }
    __device__ __forceinline__ void end() {
        // lanes finishing tasks of the same vertex (a hub's segments sit side by side in the hub queue) first sum
        // their partials, so a vertex with 10^5 segments does not serialise 10^5 fp64 atomics on one address
        cg::coalesced_group act = cg::coalesced_threads();
        cg::coalesced_group same = cg::labeled_partition(act, u);
        const double sum = cg::reduce(same, acc, cg::plus<double>());
        if (same.thread_rank() == 0 && sum != 0.0) {
            atomicAdd(delta + u, sum);
            if (u != source) atomicAdd(bc + u, sum);
        }
    }
};

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

struct CcApp {
    uint32_t* parent;
    uint32_t ru;
    uint32_t* hook_ctr;  // optional: counts successful hooks (partitioned CC convergence test)
    uint32_t hooks;
    __device__ __forceinline__ void begin(uint32_t u) {
        ru = cc_find(parent, u);
        hooks = 0;
    }
    __device__ __forceinline__ void end() {
        if (hook_ctr && hooks) atomicAdd(hook_ctr, hooks);
    }
    __device__ __forceinline__ void vertex(uint32_t) {}
    __device__ __forceinline__ void one(uint32_t v) {
        uint32_t rv = cc_find(parent, v);
        while (ru != rv) {
            const uint32_t hi = max(ru, rv), lo = min(ru, rv);
            if (atomicCAS(parent + hi, hi, lo) == hi) {
                hooks++;
                break;
            }
            ru = cc_find(parent, ru);  // hi stopped being a root: re-find both
            rv = cc_find(parent, rv);
        }
    }
    GCGT_MANY_BY_ONE
    __device__ __forceinline__ void range(uint32_t s, uint32_t len) {
        for (uint32_t t = 0; t < len; t++) one(s + t);
    }
};

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

// Direction choice for the next BFS level (Beamer et al.'s heuristic): switch to bottom-up when the new frontier is
// large against the unvisited set and growing, back to top-down when it is small against n and shrinking.
// st: [0] dir, [1] visited, [2] new-frontier count (consumed), [3] previous.  With mf_bits (record bits of the new
// frontier, summed by the contraction) the top-down -> bottom-up test is Beamer's edge form with CGR bits as the
// work measure: mf * alpha_bits > (unvisited vertices) * (mean record bits).
struct DecideArgs {
    uint32_t* st;
    uint64_t n;
    uint32_t alpha, beta;
    int enabled;
    const uint32_t* qn_len;
    uint32_t* level_counter;
    unsigned long long* mf_bits;
    double bits_per_vertex;
    uint32_t alpha_bits;
    uint32_t* done;  // blocks of commit_dense finished (the last one decides)
};

__device__ __forceinline__ void decide_body(const DecideArgs& d) {
    uint32_t* st = d.st;
    if (*(volatile const uint32_t*)d.qn_len) *d.level_counter += 1;  // levels that produced a non-empty frontier
    const uint64_t nf = *(volatile uint32_t*)(st + 2);
    st[2] = 0;
    const uint64_t visited = (uint64_t)st[1] + nf;
    st[1] = (uint32_t)visited;
    const uint64_t nu = d.n - visited, prev = st[3];
    uint32_t dir = st[0];
    bool to_bu = nf * d.alpha > nu;
    if (d.mf_bits) {
        to_bu = (double)*(volatile unsigned long long*)d.mf_bits * d.alpha_bits > (double)nu * d.bits_per_vertex;
        *d.mf_bits = 0;
    }
    if (!d.enabled || nf == 0) dir = 0;
    else if (dir == 0 && to_bu && nf > prev) dir = 1;
    else if (dir == 1 && nf * d.beta < d.n && nf < prev) dir = 0;
    st[0] = dir;
    st[3] = (uint32_t)nf;
}

// ---- contraction ---------------------------------------------------------------------------------------------------
// Dense scan of N over words [w_lo, w_hi): every non-zero word is folded into V (and F), cleared, and appended to
// the next queue (one atomic per warp).  Also resets the hub counter and the consumed queue's length.
__device__ __forceinline__ void commit_phase(uint32_t* __restrict__ V, uint32_t* __restrict__ F,
                                             uint32_t* __restrict__ N, uint64_t w_lo, uint64_t w_hi,
                                             uint32_t* __restrict__ qn, uint32_t* __restrict__ qn_len,
                                             uint32_t* __restrict__ qbits_out, int32_t* __restrict__ levels = nullptr,
                                             int32_t new_level = 0, uint32_t* __restrict__ nf_count = nullptr,
                                             const uint64_t* __restrict__ offs = nullptr,
                                             unsigned long long* __restrict__ mf_bits = nullptr) {
    const uint32_t lane = lane_id();
    const uint64_t gw = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    uint32_t nf = 0;
    uint64_t mf = 0;
    for (uint64_t base = w_lo + gw * 32; base < w_hi; base += nwarps * 32) {
        const uint64_t w = base + lane;
        uint32_t b = 0;
        if (w < w_hi) {
            b = N[w];
            if (b) {
                N[w] = 0;
                V[w] |= b;
            }
            if (F && F[w] != b) F[w] = b;  // F = exactly the new frontier
        }
        nf += __popc(b);
        if (mf_bits && b) {  // record bits of the new frontier (the top-down work estimate of bfs_decide)
            const uint64_t v0 = w * 32;
            if (b == 0xffffffffu) {
                mf += ldg64(offs + v0 + 32) - ldg64(offs + v0);
            } else {
                for (uint32_t m = b; m; m &= m - 1) {
                    const uint64_t v = v0 + __ffs(m) - 1;
                    mf += ldg64(offs + v + 1) - ldg64(offs + v);
                }
            }
        }
        const uint32_t bal = __ballot_sync(0xffffffffu, b != 0);
        if (bal) {
            uint32_t pos = 0;
            if (lane == 0) pos = atomicAdd(qn_len, __popc(bal));
            pos = __shfl_sync(0xffffffffu, pos, 0) + __popc(bal & lanemask_lt());
            if (b) {
                qn[pos] = (uint32_t)w;
                if (qbits_out) qbits_out[pos] = b;
            }
            if (levels) {  // one coalesced 32-id store per new frontier word
                for (uint32_t m = bal; m; m &= m - 1) {
                    const int j = __ffs(m) - 1;
                    const uint32_t bj = __shfl_sync(0xffffffffu, b, j);
                    if ((bj >> lane) & 1u) levels[(base + j) * 32 + lane] = new_level;
                }
            }
        }
    }
    if (nf_count) {
        for (int o = 16; o; o >>= 1) nf += __shfl_xor_sync(0xffffffffu, nf, o);
        if (lane == 0 && nf) atomicAdd(nf_count, nf);
    }
    if (mf_bits) {
        for (int o = 16; o; o >>= 1) mf += __shfl_xor_sync(0xffffffffu, mf, o);
        if (lane == 0 && mf) atomicAdd(mf_bits, (unsigned long long)mf);
    }
}

__global__ void commit_dense(uint32_t* __restrict__ V, uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                             uint64_t w_lo, uint64_t w_hi, uint32_t* __restrict__ qn, uint32_t* __restrict__ qn_len,
                             uint32_t* __restrict__ qbits_out, uint32_t* __restrict__ reset_ctr,
                             unsigned long long* __restrict__ hub_ctr, uint32_t* __restrict__ heavy_len,
                             int32_t* __restrict__ levels = nullptr, int32_t new_level = 0,
                             uint32_t* __restrict__ nf_count = nullptr,
                             unsigned long long* __restrict__ lr_ctr = nullptr,
                             const uint64_t* __restrict__ offs = nullptr,
                             unsigned long long* __restrict__ mf_bits = nullptr, DecideArgs dec = DecideArgs{}) {
    commit_phase(V, F, N, w_lo, w_hi, qn, qn_len, qbits_out, levels, new_level, nf_count, offs, mf_bits);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        if (reset_ctr) *reset_ctr = 0;
        if (hub_ctr) *hub_ctr = 0;
        if (heavy_len) *heavy_len = 0;
        if (lr_ctr) *lr_ctr = 0;
    }
    if (dec.st) {  // BFS: the last block out takes the direction decision for the next level
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            if (atomicAdd(dec.done, 1u) == gridDim.x - 1) {
                __threadfence();
                decide_body(dec);
                *dec.done = 0;
            }
        }
    }
}

// ---- bottom-up step (north_star addition; §8 a9) -----------------------------------------------------------------
// For every unvisited vertex v, decode v's IN-record until the first parent in the frontier F: intervals are tested
// as bitmap ranges (F & word mask), residuals as single bits; decoding stops at the first hit.  A warp owns one
// 32-vertex word, so the found mask is written to N without atomics.
__device__ __forceinline__ bool frontier_range(const uint32_t* __restrict__ F, uint32_t s, uint32_t len) {
    const uint32_t e = s + len;
    while (s < e) {
        const uint32_t b0 = s & 31, nb = min(32u - b0, e - s);
        if (__ldg(F + (s >> 5)) & ((nb == 32 ? 0xffffffffu : ((1u << nb) - 1)) << b0)) return true;
        s += nb;
    }
    return false;
}

// In-record scan of one unvisited vertex v: true at the first in-neighbour in F.  Residual ids are decoded four at
// a time and their four frontier probes issued together (one exit test per batch), so the probe latency is paid
// once per four arcs instead of once per arc.
template <int K, bool SEG>
__device__ __forceinline__ bool bu_scan(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                        uint32_t min_len, uint32_t seg_bits, const uint32_t* __restrict__ F,
                                        uint32_t v, uint32_t batch, uint64_t& na, uint64_t& nb) {
    const uint64_t p0 = ldg64(offs + v);
    BitBuf bb;
    bb.init(W, p0);
    uint64_t deg = 0, got = 0;
    if (!SEG) deg = bb.template next<K>(W) - 1;
    const uint64_t itv = bb.template next<K>(W) - 1;
    uint32_t prev_end = 0;
    bool found = false;
    for (uint64_t i = 0; i < itv && !found; i++) {
        const uint64_t g = bb.template next<K>(W);
        const uint32_t len = (uint32_t)(bb.template next<K>(W) - 1) + min_len;
        const uint32_t start = i == 0 ? (uint32_t)unmap_first(v, g) : prev_end + (uint32_t)g;
        found = frontier_range(F, start, len);
        prev_end = start + len - 1;
        got += len;
    }
    // residuals: cnt ids starting with one anchored at v, four per probe batch
    auto scan_res = [&](uint32_t cnt) {
        uint32_t cur = 0;
        for (uint32_t i = 0; i < cnt && !found; i += batch) {
            const uint32_t k_n = min(batch, cnt - i);
            uint32_t id[4];
#pragma unroll
            for (uint32_t k = 0; k < 4; k++) {
                if (k < k_n) {
                    const uint64_t c = bb.template next<K>(W);
                    cur = (i + k == 0) ? (uint32_t)unmap_first(v, c) : cur + (uint32_t)c;
                }
                id[k] = cur;
            }
            uint32_t fw[4];
#pragma unroll
            for (uint32_t k = 0; k < 4; k++) fw[k] = k < k_n ? __ldg(F + (id[k] >> 5)) : 0u;
#pragma unroll
            for (uint32_t k = 0; k < 4; k++) found |= ((fw[k] >> (id[k] & 31)) & 1u) != 0;
            got += k_n;
        }
    };
    uint64_t pend;
    if (found) {
        pend = bb.pos();
    } else if (!SEG) {
        scan_res((uint32_t)(deg - got));
        pend = bb.pos();
    } else {
        const uint64_t nseg = bb.template next<K>(W) - 1;
        const uint64_t base = bb.pos();
        pend = base;
        for (uint64_t sg = 0; sg < nseg && !found; sg++) {
            bb.init(W, base + sg * seg_bits);
            scan_res((uint32_t)(bb.template next<K>(W) - 1));
            pend = bb.pos();
        }
    }
    na += got;
    nb += pend - p0;
    return found;
}

// A warp owns a chunk of 8 frontier words (256 vertices): the chunk's unvisited vertices are compacted and dealt to
// the lanes round-robin (a lane per unvisited vertex, not per vertex id, so late levels with few unvisited
// vertices still fill the warp); found vertices are collected in shared memory and the warp writes its 8 words of N
// without atomics.
constexpr uint32_t kBuWords = 8;
template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock, 6) bu_kernel(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                                    uint32_t min_len, uint32_t seg_bits, const uint32_t* __restrict__ V,
                                                    const uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                                                    uint64_t n, uint64_t nw, const uint32_t* __restrict__ dir,
                                                    Stats* st, uint32_t bw, uint32_t batch,
                                                    unsigned long long* __restrict__ cur) {
    if (*dir != 1) return;
    __shared__ uint32_t found_s[kWarps][kBuWords], inc_s[kWarps][kBuWords], unv_s[kWarps][kBuWords];
    const uint32_t lane = lane_id(), wid = threadIdx.x >> 5;
    uint64_t nv = 0, na = 0, nb = 0;
    const uint64_t nch = (nw + bw - 1) / bw;
    for (;;) {
        // chunks are handed out by an atomic cursor (not grid-stride): unvisited vertices cluster, and a static
        // deal left a long tail of warps on the dense chunks (ncu, C2 level 22: 30 % warps resident, SMs idle 40 %)
        unsigned long long ch = 0;
        if (lane == 0) ch = atomicAdd(cur, 1ull);
        ch = __shfl_sync(0xffffffffu, ch, 0);
        if (ch >= nch) break;
        const uint64_t w0 = ch * bw;
        uint32_t unv = 0;
        if (lane < kBuWords) {
            found_s[wid][lane] = 0;
        }
        if (lane < bw) {
            const uint64_t w = w0 + lane, v0 = w * 32;
            if (v0 < n) {
                unv = ~__ldg(V + w);
                if (n - v0 < 32) unv &= (1u << (n - v0)) - 1;
            }
        }
        uint32_t cnt = lane < kBuWords ? __popc(unv) : 0, incl = cnt;
        for (int o = 1; o < (int)kBuWords; o <<= 1) {
            const uint32_t t = __shfl_up_sync(0xffffffffu, incl, o);
            if (lane >= (uint32_t)o) incl += t;
        }
        const uint32_t total = __shfl_sync(0xffffffffu, incl, kBuWords - 1);
        if (!total) continue;
        if (lane < kBuWords) {
            inc_s[wid][lane] = incl;
            unv_s[wid][lane] = unv;
        }
        __syncwarp();
        for (uint32_t r = lane; r < total; r += 32) {
            // candidate r: word k with excl(k) <= r < incl(k)
            uint32_t k = 0, ex = 0, bits = 0;
#pragma unroll
            for (uint32_t q = 0; q < kBuWords; q++) {
                const uint32_t iq = inc_s[wid][q], bq = unv_s[wid][q];
                const uint32_t eq = iq - __popc(bq);
                if (r >= eq && r < iq) { k = q; ex = eq; bits = bq; }
            }
            const uint32_t bit = __fns(bits, 0, (int)(r - ex) + 1);
            const uint32_t v = (uint32_t)((w0 + k) * 32 + bit);
            nv++;
            if (bu_scan<K, SEG>(W, offs, min_len, seg_bits, F, v, batch, na, nb)) atomicOr(&found_s[wid][k], 1u << bit);
        }
        __syncwarp();
        if (lane < kBuWords) {
            const uint32_t m = found_s[wid][lane];
            if (m) N[w0 + lane] = m;
        }
        __syncwarp();
    }
    add_stats(st, nv, na, nb);
    __syncthreads();
    if (threadIdx.x == 0 && atomicAdd(cur + 1, 1ull) == gridDim.x - 1) {  // last block out resets the cursor
        cur[0] = 0;
        cur[1] = 0;
    }
}

// Per-word variant (round 1): lane = vertex of the warp's 32-vertex word, one frontier probe per residual.
template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock) bu_kernel1(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs,
                                                    uint32_t min_len, uint32_t seg_bits, const uint32_t* __restrict__ V,
                                                    const uint32_t* __restrict__ F, uint32_t* __restrict__ N,
                                                    uint64_t n, uint64_t nw, const uint32_t* __restrict__ dir,
                                                    Stats* st) {
    if (*dir != 1) return;
    const uint32_t lane = lane_id();
    uint64_t nv = 0, na = 0, nb = 0;
    for (uint64_t w = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5; w < nw;
         w += ((uint64_t)gridDim.x * blockDim.x) >> 5) {
        const uint64_t v0 = w * 32;
        if (v0 >= n) break;
        uint32_t unv = ~__ldg(V + w);
        if (n - v0 < 32) unv &= (1u << (n - v0)) - 1;
        if (!unv) continue;
        bool found = false;
        if ((unv >> lane) & 1u) {
            // BitBuf decoding: this kernel is instruction-bound (long in-record scans at high lane utilisation), so
            // the cheaper 32-bit refill decoder pays off here (unlike the latency-bound top-down kernel)
            const uint32_t v = (uint32_t)(v0 + lane);
            const uint64_t p0 = ldg64(offs + v);
            BitBuf bb;
            bb.init(W, p0);
            nv++;
            uint64_t deg = 0, got = 0, pend = p0;
            if (!SEG) deg = bb.template next<K>(W) - 1;
            const uint64_t itv = bb.template next<K>(W) - 1;
            uint32_t prev_end = 0;
            for (uint64_t i = 0; i < itv && !found; i++) {
                const uint64_t g = bb.template next<K>(W);
                const uint32_t len = (uint32_t)(bb.template next<K>(W) - 1) + min_len;
                const uint32_t start = i == 0 ? (uint32_t)unmap_first(v, g) : prev_end + (uint32_t)g;
                found = frontier_range(F, start, len);
                prev_end = start + len - 1;
                got += len;
            }
            if (!found) {
                if (!SEG) {
                    const uint64_t nres = deg - got;
                    uint32_t cur = 0;
                    for (uint64_t i = 0; i < nres && !found; i++) {
                        const uint64_t c = bb.template next<K>(W);
                        cur = i == 0 ? (uint32_t)unmap_first(v, c) : cur + (uint32_t)c;
                        found = (__ldg(F + (cur >> 5)) >> (cur & 31)) & 1u;
                        got++;
                    }
                    pend = bb.pos();
                } else {
                    const uint64_t nseg = bb.template next<K>(W) - 1;
                    const uint64_t base = bb.pos();
                    pend = base;
                    for (uint64_t sg = 0; sg < nseg && !found; sg++) {
                        bb.init(W, base + sg * seg_bits);
                        const uint32_t cnt = (uint32_t)(bb.template next<K>(W) - 1);
                        uint32_t cur = 0;
                        for (uint32_t i = 0; i < cnt && !found; i++) {
                            const uint64_t c = bb.template next<K>(W);
                            cur = i == 0 ? (uint32_t)unmap_first(v, c) : cur + (uint32_t)c;
                            found = (__ldg(F + (cur >> 5)) >> (cur & 31)) & 1u;
                            got++;
                        }
                        pend = bb.pos();
                    }
                }
            } else {
                pend = bb.pos();
            }
            na += got;
            nb += pend - p0;
        }
        const uint32_t fb = __ballot_sync(0xffffffffu, found);
        if (lane == 0 && fb) N[w] = fb;
    }
    add_stats(st, nv, na, nb);
}

// ---- persistent BFS: every level inside one cooperative launch ------------------------------------------------------
// Per level: expansion (work cursor) | grid sync | hub segments | grid sync | contraction into the next queue |
// grid sync.  No host round trip per level: the host launches once and waits once (high-diameter web graphs have
// dozens of levels, and each host-driven level costs launches plus a stream synchronisation).
struct BfsPersist {
    uint32_t* q0;
    uint32_t* q1;
    uint32_t* ctr;     // [0], [1]: queue lengths (ping-pong); [6]: levels expanded (out)
    uint32_t* V;
    uint32_t* F;
    uint32_t* N;
    int32_t* levels;
    uint64_t nw;
    uint32_t wpb_max;
};

template <int K, bool SEG>
__global__ void __launch_bounds__(kBlock, 4) bfs_persistent(Ctx c, BfsPersist b) {
    __shared__ WarpSmem smem[kWarps];
    cg::grid_group grid = cg::this_grid();
    uint64_t nv = 0, na = 0, nb = 0;
    const uint64_t nwarps = (uint64_t)gridDim.x * kWarps;
    uint32_t level = 0;
    for (;; level++) {
        const int cur = level & 1, nxt = cur ^ 1;
        uint32_t* qc = cur ? b.q1 : b.q0;
        uint32_t* qn = cur ? b.q0 : b.q1;
        const uint64_t qlen = *(volatile uint32_t*)(b.ctr + cur);
        uint64_t wpb = qlen / (nwarps * 4);
        wpb = wpb < 1 ? 1 : (wpb > b.wpb_max ? b.wpb_max : wpb);
        const QueueFront fr{qc, b.ctr + cur, b.F, nullptr};
        const BfsApp app{b.V, b.N, b.levels, (int32_t)level};
        expand_phase<K, SEG, BfsApp, QueueFront, true, false>(c, fr, app, (uint32_t)wpb, smem, nv, na, nb);
        grid.sync();
        if (SEG || c.hv_n || c.lr_ctr) {
            hub_phase<K, false>(c, app, na);
            grid.sync();
        }
        commit_phase(b.V, b.F, b.N, 0, b.nw, qn, b.ctr + nxt, nullptr, b.levels, (int32_t)level + 1);
        if (blockIdx.x == 0 && threadIdx.x == 0) {
            b.ctr[cur] = 0;
            *c.hub_ctr = 0;
            if (c.lr_ctr) *c.lr_ctr = 0;
            c.cursor[0] = 0;
        }
        grid.sync();
        if (*(volatile uint32_t*)(b.ctr + nxt) == 0) break;
    }
    add_stats(c.st, nv, na, nb);
    if (blockIdx.x == 0 && threadIdx.x == 0) b.ctr[6] = level + 1;
}

// ---- partitioned BFS / CC steps (the collectives run in the caller, e.g. torch.distributed over NCCL) ------------
// Contraction of the owned slice: OR of the P candidate slices received from every rank, minus visited; writes
// levels and the owned next-frontier slice; counts new vertices.
__global__ void dist_commit(const uint32_t* __restrict__ recv, uint32_t P, uint64_t w_lo, uint64_t nlw,
                            const uint32_t* __restrict__ V, uint32_t* __restrict__ fslice, int32_t* __restrict__ levels,
                            int32_t new_level, uint64_t n, unsigned long long* __restrict__ count) {
    const uint32_t lane = lane_id();
    uint32_t nf = 0;
    const uint64_t gw = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    for (uint64_t base = gw * 32; base < nlw; base += nwarps * 32) {
        const uint64_t i = base + lane;
        uint32_t b = 0;
        if (i < nlw) {
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

// F = the gathered global frontier; V |= F.
__global__ void dist_absorb(const uint32_t* __restrict__ Fg, uint32_t* __restrict__ F, uint32_t* __restrict__ V,
                            uint64_t nw) {
    for (uint64_t w = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; w < nw; w += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t b = Fg[w];
        F[w] = b;
        V[w] |= b;
    }
}

__global__ void bfs_seed(uint32_t s, uint32_t* V, uint32_t* F, uint32_t* q, uint32_t* qlen, uint32_t* qbits,
                         int32_t* levels = nullptr, uint32_t* bstate = nullptr) {
    V[s >> 5] = 1u << (s & 31);
    if (levels) levels[s] = 0;
    if (bstate) {
        bstate[0] = 0;
        bstate[1] = 1;
        bstate[2] = 0;
        bstate[3] = 1;
    }
    if (F) F[s >> 5] = 1u << (s & 31);
    q[0] = s >> 5;
    if (qbits) qbits[0] = 1u << (s & 31);
    *qlen = 1;
}

__global__ void bswap_words(uint64_t* w, uint64_t n) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x)
        w[i] = __byte_perm((uint32_t)(w[i] >> 32), 0, 0x0123) | ((uint64_t)__byte_perm((uint32_t)w[i], 0, 0x0123) << 32);
}

// ---- load-time interval checkpoint table ---------------------------------------------------------------------------
// Vertices with more than C intervals get a checkpoint every C intervals: the bit position of the gap code of
// interval kC and the end of interval kC-1.  Each chunk of C intervals then decodes on its own, so a long interval
// area no longer forms one serial chain (the residual-segment idea of §5.2 applied to intervals, as a derived
// device table; the CGR bytes are unchanged).
template <int K, bool SEG>
__global__ void ck_count(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs, uint64_t lo, uint64_t n,
                         uint32_t C, uint8_t* __restrict__ flag, uint32_t* __restrict__ cnt) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint64_t u = lo + i;  // flag / cnt are indexed by owned position; the selected ids are re-based below
        uint64_t p = ldg64(offs + u);
        if (!SEG) decode<K>(W, p);
        const uint64_t itv = decode<K>(W, p) - 1;
        const bool h = itv > C;
        flag[i] = h;
        cnt[i] = h ? (uint32_t)((itv - 1) / C) : 0;
    }
}

// Per-word index of the checkpoint table: wptr[w - w0] = number of table vertices below 32w, bits[w - w0] = which
// of the word's 32 vertices are in the table.  A frontier vertex finds its table row with two independent loads
// instead of a ~17-step dependent binary search over the sorted ids (the tail levels' critical path).
__global__ void hv_index(const uint32_t* __restrict__ ids, uint32_t H, uint64_t w0, uint64_t nwl,
                         uint32_t* __restrict__ wptr, uint32_t* __restrict__ bits) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i <= nwl; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint64_t v0 = (w0 + i) * 32;
        uint32_t lo = 0, hi = H;
        while (lo < hi) {
            const uint32_t mid = (lo + hi) >> 1;
            if (ids[mid] < v0) lo = mid + 1; else hi = mid;
        }
        wptr[i] = lo;
        uint32_t b = 0;
        for (uint32_t j = lo; j < H && ids[j] < v0 + 32; j++) b |= 1u << (ids[j] - v0);
        if (i < nwl) bits[i] = b;
    }
}

__global__ void ck_gather(uint32_t* __restrict__ ids, const uint32_t* __restrict__ cnt, uint32_t H, uint64_t lo,
                          uint32_t* __restrict__ out) {
    for (uint64_t h = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; h <= H; h += (uint64_t)gridDim.x * blockDim.x) {
        out[h] = h < H ? cnt[ids[h]] : 0;
        if (h < H) ids[h] += (uint32_t)lo;  // owned position -> global vertex id
    }
}

template <int K, bool SEG>
__global__ void ck_fill(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs, uint32_t min_len,
                        uint32_t C, const uint32_t* __restrict__ ids, const uint32_t* __restrict__ ptr, uint32_t H,
                        uint64_t* __restrict__ ck_pos, uint32_t* __restrict__ ck_prev, uint64_t* __restrict__ after,
                        uint32_t* __restrict__ rem) {
    for (uint64_t h = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; h < H; h += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t u = ids[h];
        uint64_t p = ldg64(offs + u), deg = 0, sum = 0;
        if (!SEG) deg = decode<K>(W, p) - 1;
        const uint64_t itv = decode<K>(W, p) - 1;
        int64_t prev_end = 0;
        for (uint64_t i = 0; i < itv; i++) {
            if (i && i % C == 0) {
                const uint32_t k = ptr[h] + (uint32_t)(i / C) - 1;
                ck_pos[k] = p;
                ck_prev[k] = (uint32_t)prev_end;
            }
            const uint64_t g = decode<K>(W, p);
            const uint64_t len = decode<K>(W, p) - 1 + min_len;
            const int64_t start = i == 0 ? unmap_first(u, g) : prev_end + (int64_t)g;
            prev_end = start + (int64_t)len - 1;
            sum += len;
        }
        after[h] = p;
        rem[h] = SEG ? 0 : (uint32_t)(deg - sum);
    }
}

// Load-time pass: number of hub vertices (more than kHubSegs residual segments) and heavy vertices (long
// interval area / unsegmented list); sizes the per-level hub and heavy queues.
template <int K, bool SEG>
__global__ void count_special(const uint64_t* __restrict__ W, const uint64_t* __restrict__ offs, uint64_t lo,
                              uint64_t n, uint32_t heavy_itv, uint32_t heavy_res, uint32_t hub_segs,
                              uint32_t min_len, uint32_t long_len, unsigned long long* out) {
    uint32_t hubs = 0, heavy = 0, longs = 0;
    for (uint64_t u = lo + (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; u < n;
         u += (uint64_t)gridDim.x * blockDim.x) {
        uint64_t p = ldg64(offs + u);
        uint64_t deg = 0;
        if (!SEG) deg = decode<K>(W, p) - 1;
        const uint64_t itv = decode<K>(W, p) - 1;
        if (itv > heavy_itv || (!SEG && deg > heavy_res)) heavy++;
        for (uint64_t i = 0; i < itv; i++) {
            decode<K>(W, p);
            if (decode<K>(W, p) - 1 + min_len > long_len) longs++;
        }
        if (SEG && decode<K>(W, p) - 1 > hub_segs) hubs++;
    }
    for (int o = 16; o; o >>= 1) {
        hubs += __shfl_xor_sync(0xffffffffu, hubs, o);
        heavy += __shfl_xor_sync(0xffffffffu, heavy, o);
        longs += __shfl_xor_sync(0xffffffffu, longs, o);
    }
    if (lane_id() == 0) {
        if (hubs) atomicAdd(out, (unsigned long long)hubs);
        if (heavy) atomicAdd(out + 1, (unsigned long long)heavy);
        if (longs) atomicAdd(out + 2, (unsigned long long)longs);
    }
}

// ---- dispatch -------------------------------------------------------------------------------------------------------
// Persistent launch: at most one wave (occupancy calculator), never more blocks than the work needs.
template <int K, bool SEG, class App, class Front, bool DEFER, bool STAGED>
inline void launch_expand_k(int grid, cudaStream_t s, const Ctx& c, const Front& fr, const App& app, uint32_t wpb) {
    static int sms = 0;
    if (!sms) {
        int dev = 0;
        cudaGetDevice(&dev);
        cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    }
    if (DEFER && c.engine == 1) {  // state-machine kernel (default); no heavy deferral needed
        static int per_sm = 0;
        if (!per_sm) {
            cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, sm_expand_kernel<K, SEG, App, Front>, kBlock, 0);
            if (per_sm < 1) per_sm = 1;
        }
        grid = std::max(1, std::min(grid, per_sm * sms));
        sm_expand_kernel<K, SEG, App, Front><<<grid, kBlock, 0, s>>>(c, fr, app, wpb);
        return;
    }
    static int per_sm = 0;
    if (!per_sm) {
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, expand_kernel<K, SEG, App, Front, DEFER, STAGED>, kBlock,
                                                      0);
        if (per_sm < 1) per_sm = 1;
    }
    grid = std::max(1, std::min(grid, per_sm * sms));
    expand_kernel<K, SEG, App, Front, DEFER, STAGED><<<grid, kBlock, 0, s>>>(c, fr, app, wpb);
}

template <class App, class Front, bool DEFER = true>
inline void launch_expand(const gcgt_params& P, bool staged, int grid, cudaStream_t s, const Ctx& c,
                          const Front& fr, const App& app, uint32_t wpb) {
    const bool seg = P.residual_segment_len != 0;
#define GCGT_EXP(KK)                                                                                          \
    (staged ? (seg ? launch_expand_k<KK, true, App, Front, DEFER, true>(grid, s, c, fr, app, wpb)              \
                   : launch_expand_k<KK, false, App, Front, DEFER, true>(grid, s, c, fr, app, wpb))            \
            : (seg ? launch_expand_k<KK, true, App, Front, DEFER, false>(grid, s, c, fr, app, wpb)             \
                   : launch_expand_k<KK, false, App, Front, DEFER, false>(grid, s, c, fr, app, wpb)))
    switch (P.zeta_k) {
        case 1: GCGT_EXP(1); break;
        case 2: GCGT_EXP(2); break;
        case 3: GCGT_EXP(3); break;
        case 4: GCGT_EXP(4); break;
        default: GCGT_EXP(5); break;
    }
#undef GCGT_EXP
}

// Heavy pass: the same engine over the level's heavy queue, 32 heavy vertices per warp batch.
inline bool heavy_active(const gcgt_graph* g) {  // can any vertex be deferred to the heavy pass?
    if (g->engine == 1) return false;                  // the state-machine kernel never defers
    return g->heavy_itv != 0xFFFFFFFFu || (g->P.residual_segment_len == 0 && g->heavy_res != 0xFFFFFFFFu);
}

template <class App>
inline void launch_heavy(const gcgt_graph* g, cudaStream_t s, const Ctx& c, const App& app) {
    if (!heavy_active(g)) return;
    const HeavyFront fr{c.heavyq, c.heavy_len};
    launch_expand<App, HeavyFront, false>(g->P, g->staged, g->num_sms * 8, s, c, fr, app, 32);
}

// Cooperative launch of the persistent BFS (one wave, co-resident blocks).  Returns false if the device cannot
// co-schedule the grid (then the host-driven level loop is used).
template <int K, bool SEG>
inline cudaError_t launch_bfs_persistent_k(const gcgt_graph* g, cudaStream_t s, Ctx c, BfsPersist b) {
    static int per_sm = -1;
    if (per_sm < 0) {
        if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, bfs_persistent<K, SEG>, kBlock, 0) != cudaSuccess)
            per_sm = 0;
    }
    if (per_sm < 1) return cudaErrorCooperativeLaunchTooLarge;
    void* args[] = {(void*)&c, (void*)&b};
    return cudaLaunchCooperativeKernel((const void*)bfs_persistent<K, SEG>, dim3(per_sm * g->num_sms), dim3(kBlock),
                                       args, 0, s);
}

inline cudaError_t launch_bfs_persistent(const gcgt_graph* g, cudaStream_t s, Ctx c, const BfsPersist& b) {
    c.heavy_itv = 0xFFFFFFFFu;  // nothing is deferred inside the persistent loop
    c.heavy_res = 0xFFFFFFFFu;
    const bool seg = g->P.residual_segment_len != 0;
    switch (g->P.zeta_k) {
        case 1: return seg ? launch_bfs_persistent_k<1, true>(g, s, c, b) : launch_bfs_persistent_k<1, false>(g, s, c, b);
        case 2: return seg ? launch_bfs_persistent_k<2, true>(g, s, c, b) : launch_bfs_persistent_k<2, false>(g, s, c, b);
        case 3: return seg ? launch_bfs_persistent_k<3, true>(g, s, c, b) : launch_bfs_persistent_k<3, false>(g, s, c, b);
        case 4: return seg ? launch_bfs_persistent_k<4, true>(g, s, c, b) : launch_bfs_persistent_k<4, false>(g, s, c, b);
        default: return seg ? launch_bfs_persistent_k<5, true>(g, s, c, b) : launch_bfs_persistent_k<5, false>(g, s, c, b);
    }
}

template <int K, bool SEG>
inline void launch_bu_k(const gcgt_graph* g, cudaStream_t s) {
    static int per_sm = 0, per_sm1 = 0;
    if (!per_sm) {
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, bu_kernel<K, SEG>, kBlock, 0);
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm1, bu_kernel1<K, SEG>, kBlock, 0);
        if (per_sm < 1) per_sm = 1;
        if (per_sm1 < 1) per_sm1 = 1;
    }
    if (g->bu_kernel == 1) {  // round-1 per-word kernel
        const int grid = (int)std::max<uint64_t>(1, std::min<uint64_t>((g->nw + kWarps - 1) / kWarps,
                                                                        (uint64_t)per_sm1 * g->num_sms));
        bu_kernel1<K, SEG><<<grid, kBlock, 0, s>>>(g->inW, g->inOffs, g->P.min_interval_len,
                                                   8 * g->P.residual_segment_len, g->V, g->F, g->N, g->n, g->nw,
                                                   g->bstate, g->stats);
        return;
    }
    const uint64_t chunks = (g->nw + g->bu_words - 1) / g->bu_words;
    const int grid = (int)std::max<uint64_t>(1, std::min<uint64_t>((chunks + kWarps - 1) / kWarps,
                                                                    (uint64_t)per_sm * g->num_sms));
    bu_kernel<K, SEG><<<grid, kBlock, 0, s>>>(g->inW, g->inOffs, g->P.min_interval_len, 8 * g->P.residual_segment_len,
                                              g->V, g->F, g->N, g->n, g->nw, g->bstate, g->stats,
                                              g->bu_words, g->bu_batch, g->bu_cur);
}

inline void launch_bu(const gcgt_graph* g, cudaStream_t s) {
    const bool seg = g->P.residual_segment_len != 0;
    switch (g->P.zeta_k) {
        case 1: seg ? launch_bu_k<1, true>(g, s) : launch_bu_k<1, false>(g, s); break;
        case 2: seg ? launch_bu_k<2, true>(g, s) : launch_bu_k<2, false>(g, s); break;
        case 3: seg ? launch_bu_k<3, true>(g, s) : launch_bu_k<3, false>(g, s); break;
        case 4: seg ? launch_bu_k<4, true>(g, s) : launch_bu_k<4, false>(g, s); break;
        default: seg ? launch_bu_k<5, true>(g, s) : launch_bu_k<5, false>(g, s); break;
    }
}

// The hub pass is latency-bound (one segment's dependent codeword chain per thread): launch a full wave at the
// kernel's occupancy rather than a fixed 4 blocks per SM (`grid` = 4 blocks per SM is the floor).
template <int K, bool STAGED, class App>
inline int hub_wave(int grid) {
    static int wave = 0;
    if (!wave) {
        int dev = 0, sms = 0, per_sm = 0;
        cudaGetDevice(&dev);
        cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, hub_kernel<K, STAGED, App>, kBlock, 0);
        wave = std::max(1, per_sm) * std::max(1, sms);
    }
    return std::max(grid, wave);
}

template <class App>
inline void launch_hub(const gcgt_params& P, bool staged, int grid, cudaStream_t s, const Ctx& c, const App& app) {
    if (c.fuse) return;  // drained inside expand_kernel
    if (!P.residual_segment_len && !c.hv_n && !c.lr_ctr) return;
    (void)staged;  // hub segments always use the BitBuf reader (C3: hub pass 1.40 vs 2.05 ms; C2 unchanged)
#define GCGT_HUB(KK) hub_kernel<KK, true, App><<<hub_wave<KK, true, App>(grid), kBlock, 0, s>>>(c, app)
    switch (P.zeta_k) {
        case 1: GCGT_HUB(1); break;
        case 2: GCGT_HUB(2); break;
        case 3: GCGT_HUB(3); break;
        case 4: GCGT_HUB(4); break;
        default: GCGT_HUB(5); break;
    }
#undef GCGT_HUB
}

// Work granularity for a frontier of qlen words: every resident warp should take several batches (dynamic
// balancing); small frontiers get one word per batch and only as many blocks as there are words.
inline void frontier_launch(const gcgt_graph* g, uint64_t qlen, int* grid, uint32_t* wpb) {
    const uint64_t resident_warps = (uint64_t)g->num_sms * 48;
    uint64_t b = qlen / (resident_warps * 4);
    b = std::max<uint64_t>(1, std::min<uint64_t>(b, g->wpb_max));
    const uint64_t warps = (qlen + b - 1) / b;
    *grid = (int)std::max<uint64_t>(1, std::min<uint64_t>((warps + kWarps - 1) / kWarps, (uint64_t)g->num_sms * 32));
    *wpb = (uint32_t)b;
}

inline int flat_grid(const gcgt_graph* g, uint64_t n) {
    return (int)std::max<uint64_t>(1, std::min<uint64_t>((n + kBlock - 1) / kBlock, (uint64_t)g->num_sms * 16));
}

inline int hub_grid(const gcgt_graph* g) { return g->num_sms * 4; }

inline Ctx make_ctx(const gcgt_graph* g) {
    return Ctx{g->W,     g->offs,     g->P.min_interval_len, 8 * g->P.residual_segment_len,
               g->hubq, g->hub_ctr, g->stats,              g->cursor,
               g->heavyq, g->heavy_len, g->heavy_itv, g->heavy_res, g->hub_segs, g->engine, nullptr,
               g->hv_n,  g->ck_c,      g->hv_ids,    g->hv_ptr,    g->hv_wptr, g->hv_bits, g->lo >> 5, g->hv_after, g->hv_rem, g->ck_pos, g->ck_prev,
               g->lrq,   g->lr_ctr,    g->long_len,  g->lr_chunk,
               (!heavy_active(g) && g->engine == 0 && g->fuse_ctr) ? g->fuse_warps : 0u, g->fuse_ctr, g->flatb};
}

gcgt_status copy_out(gcgt_graph* g, void* dst, const void* src, size_t bytes, int placement) {
    CU(cudaMemcpyAsync(dst, src, bytes, placement == GCGT_OUT_DEVICE ? cudaMemcpyDeviceToDevice : cudaMemcpyDeviceToHost,
                       g->stream));
    return GCGT_OK;
}

#include "csr_bfs.cuh"

// Brackets one launch of the dominant kernel when profiling (the caller syncs before reading).
// Profiled launches record into a pool of event pairs (created on first use) and are read at the next host sync,
// so timing does not force a per-level wait (the chunked BFS level loop keeps its asynchronous enqueue).
inline gcgt_status kprof_begin(gcgt_graph* g) {
    if (!g->profile) return GCGT_OK;
    if (g->kev_n >= gcgt_graph::kKev) return fail(GCGT_EINVAL, "too many profiled launches between syncs");
    cudaEvent_t& e = g->kevp[2 * g->kev_n];
    if (!e) CU(cudaEventCreate(&e));
    CU(cudaEventRecord(e, g->stream));
    return GCGT_OK;
}
inline gcgt_status kprof_end(gcgt_graph* g) {
    if (!g->profile) return GCGT_OK;
    cudaEvent_t& e = g->kevp[2 * g->kev_n + 1];
    if (!e) CU(cudaEventCreate(&e));
    CU(cudaEventRecord(e, g->stream));
    g->kev_n++;
    return GCGT_OK;
}
inline gcgt_status kprof_collect(gcgt_graph* g) {  // after a stream sync
    if (!g->profile) return GCGT_OK;
    for (int i = 0; i < g->kev_n; i++) {
        float ms = 0;
        CU(cudaEventElapsedTime(&ms, g->kevp[2 * i], g->kevp[2 * i + 1]));
        g->kernel_ms += ms;
        g->kernel_launches++;
    }
    g->kev_n = 0;
    return GCGT_OK;
}

gcgt_status begin_call(gcgt_graph* g) {
    gcgt_internal::clear_error();
    CU(cudaSetDevice(g->device));
    g->kernel_ms = 0;
    g->kernel_launches = 0;
    g->launches = 0;
    for (double& x : g->span_ms) x = 0;
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
        out->launches = g->launches;
    }
    return GCGT_OK;
}

// Small pinned host blocks (per-graph counters and stats) are recycled process-wide: cudaFreeHost on every unload
// measured 0.6 ms typical with stalls of 12-314 ms (tools/e2e_breakdown.py, session 4), inside the e2e step.
static constexpr size_t kSmallPinned = 256;
static std::mutex g_small_mu;
static std::vector<void*> g_small_free;
static cudaError_t small_pinned_get(void** p) {
    {
        std::lock_guard<std::mutex> lk(g_small_mu);
        if (!g_small_free.empty()) {
            *p = g_small_free.back();
            g_small_free.pop_back();
            return cudaSuccess;
        }
    }
    return cudaMallocHost(p, kSmallPinned);
}
static void small_pinned_put(void* p) {
    if (!p) return;
    std::lock_guard<std::mutex> lk(g_small_mu);
    g_small_free.push_back(p);
}
static_assert(sizeof(Stats) <= kSmallPinned && 8 * sizeof(uint32_t) <= kSmallPinned, "small pinned block size");

// Wall-clock marks of load / unload phases on stderr when GCGT_TIMING is set (diagnostics for the bench's e2e leg).
struct PhaseClock {
    bool on = getenv("GCGT_TIMING") != nullptr;
    const char* what;
    std::chrono::steady_clock::time_point t0 = std::chrono::steady_clock::now(), t = t0;
    explicit PhaseClock(const char* w) : what(w) {}
    void mark(const char* phase, cudaStream_t s = nullptr) {
        if (!on) return;
        if (s) cudaStreamSynchronize(s);
        const auto now = std::chrono::steady_clock::now();
        fprintf(stderr, "[%s] %-18s %8.2f ms (total %8.2f)\n", what, phase,
                std::chrono::duration<double, std::milli>(now - t).count(),
                std::chrono::duration<double, std::milli>(now - t0).count());
        t = now;
    }
};

template <class T>
gcgt_status dalloc(T** p, uint64_t count) {
    cudaError_t e = cudaMalloc((void**)p, std::max<uint64_t>(1, count) * sizeof(T));
    if (e != cudaSuccess) return fail(GCGT_ENOMEM, std::string("cudaMalloc: ") + cudaGetErrorString(e));
    return GCGT_OK;
}

// Graph buffers come from the device's stream-ordered memory pool, which keeps freed memory (release threshold =
// max), so repeated load / unload cycles (the bench's end-to-end leg, query services) reuse device memory instead
// of paying cudaMalloc / cudaFree each time.
template <class T>
gcgt_status galloc(const gcgt_graph* g, T** p, uint64_t count) {
    cudaError_t e = cudaMallocAsync((void**)p, std::max<uint64_t>(1, count) * sizeof(T), g->stream);
    if (e != cudaSuccess) return fail(GCGT_ENOMEM, std::string("cudaMallocAsync: ") + cudaGetErrorString(e));
    return GCGT_OK;
}

}  // namespace

// Host-resident CGR words (§8 f4): a pinned, mapped host buffer holding words [w0, w0 + nwords) of the canonical
// stream, byte-swapped on the host into the device's stream-word order; *dev is its device alias.  The kernels then
// decode straight from host memory over the host link (the paper's out-of-core motivation, PAPER.md:93-120,
// :474-479: graphs whose CGR exceeds device memory), while every O(n) table stays in HBM.
gcgt_status host_words(gcgt_graph* g, uint64_t** host, uint64_t** dev, const std::vector<uint64_t>& words,
                       uint64_t w0, uint64_t nwords) {
    (void)g;
    CU(cudaHostAlloc((void**)host, nwords * sizeof(uint64_t), cudaHostAllocMapped | cudaHostAllocPortable));
    uint64_t* h = *host;
    const uint64_t avail = words.size() > w0 ? words.size() - w0 : 0;
#pragma omp parallel for schedule(static)
    for (int64_t i = 0; i < (int64_t)nwords; i++)
        h[i] = (uint64_t)i < avail ? __builtin_bswap64(words[w0 + i]) : 0;
    CU(cudaHostGetDevicePointer((void**)dev, h, 0));
    return GCGT_OK;
}

// Builds the interval checkpoint table (see ck_count / ck_fill) and the per-level chunk queue.
gcgt_status build_checkpoints(gcgt_graph* g) {
    gcgt_status st;
    if ((st = galloc(g, &g->lr_ctr, 1))) return st;
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, g->stream));
    if (g->ck_c == 0xFFFFFFFFu || g->hi == g->lo) return GCGT_OK;
    cudaStream_t s = g->stream;
    const bool seg = g->P.residual_segment_len != 0;
    const uint32_t C = g->ck_c;
    uint8_t* flag = nullptr;
    uint32_t *cnt = nullptr, *ids = nullptr, *nsel = nullptr;
    if ((st = galloc(g, &flag, g->hi - g->lo + 1)) || (st = galloc(g, &cnt, g->hi - g->lo + 1)) ||
        (st = galloc(g, &ids, g->hi - g->lo + 1)) ||
        (st = galloc(g, &nsel, 1)))
        return st;
    const uint64_t nloc = g->hi - g->lo;
    const int gr = flat_grid(g, nloc);
#define GCGT_CK(KK) (seg ? ck_count<KK, true><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, nloc, C, flag, cnt)   \
                         : ck_count<KK, false><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, nloc, C, flag, cnt))
    switch (g->P.zeta_k) {
        case 1: GCGT_CK(1); break;
        case 2: GCGT_CK(2); break;
        case 3: GCGT_CK(3); break;
        case 4: GCGT_CK(4); break;
        default: GCGT_CK(5); break;
    }
#undef GCGT_CK
    size_t tmp_bytes = 0;
    cub::CountingInputIterator<uint32_t> iota(0);
    CU(cub::DeviceSelect::Flagged(nullptr, tmp_bytes, iota, flag, ids, nsel, (int64_t)nloc, s));
    void* tmp = nullptr;
    size_t tmp2 = 0;
    CU(cub::DeviceScan::ExclusiveSum(nullptr, tmp2, cnt, cnt, (int64_t)nloc + 1, s));
    if ((st = galloc(g, (uint8_t**)&tmp, std::max(tmp_bytes, tmp2)))) return st;
    CU(cub::DeviceSelect::Flagged(tmp, tmp_bytes, iota, flag, ids, nsel, (int64_t)nloc, s));
    uint32_t H = 0;
    CU(cudaMemcpyAsync(&H, nsel, 4, cudaMemcpyDeviceToHost, s));
    CU(cudaStreamSynchronize(s));
    if (H) {
        if ((st = galloc(g, &g->hv_ids, H)) || (st = galloc(g, &g->hv_ptr, H + 1)) ||
            (st = galloc(g, &g->hv_after, H)) || (st = galloc(g, &g->hv_rem, H)))
            return st;
        CU(cudaMemcpyAsync(g->hv_ids, ids, (uint64_t)H * 4, cudaMemcpyDeviceToDevice, s));
        ck_gather<<<flat_grid(g, H + 1), kBlock, 0, s>>>(g->hv_ids, cnt, H, g->lo, ids);
        // ids now holds the per-heavy-vertex counts (+ a trailing 0); scan into hv_ptr
        tmp2 = std::max(tmp_bytes, tmp2);
        CU(cub::DeviceScan::ExclusiveSum(tmp, tmp2, ids, g->hv_ptr, (int64_t)H + 1, s));
        uint32_t T = 0;
        CU(cudaMemcpyAsync(&T, g->hv_ptr + H, 4, cudaMemcpyDeviceToHost, s));
        CU(cudaStreamSynchronize(s));
        if ((st = galloc(g, &g->ck_pos, (uint64_t)T + 1)) || (st = galloc(g, &g->ck_prev, (uint64_t)T + 1)))
            return st;
        const int gh = flat_grid(g, H);
#define GCGT_CF(KK)                                                                                                  \
    (seg ? ck_fill<KK, true><<<gh, kBlock, 0, s>>>(g->W, g->offs, g->P.min_interval_len, C, g->hv_ids, g->hv_ptr, H, \
                                                   g->ck_pos, g->ck_prev, g->hv_after, g->hv_rem)                      \
         : ck_fill<KK, false><<<gh, kBlock, 0, s>>>(g->W, g->offs, g->P.min_interval_len, C, g->hv_ids, g->hv_ptr,  \
                                                    H, g->ck_pos, g->ck_prev, g->hv_after, g->hv_rem))
        switch (g->P.zeta_k) {
            case 1: GCGT_CF(1); break;
            case 2: GCGT_CF(2); break;
            case 3: GCGT_CF(3); break;
            case 4: GCGT_CF(4); break;
            default: GCGT_CF(5); break;
        }
#undef GCGT_CF
        g->hv_n = H;
        const uint64_t w0 = g->lo >> 5, nwl = ((g->hi + 31) >> 5) - w0;
        if ((st = galloc(g, &g->hv_wptr, nwl + 1)) || (st = galloc(g, &g->hv_bits, nwl + 1))) return st;
        hv_index<<<flat_grid(g, nwl + 1), kBlock, 0, s>>>(g->hv_ids, H, w0, nwl, g->hv_wptr, g->hv_bits);
    }
    cudaFreeAsync(flag, s);
    cudaFreeAsync(cnt, s);
    cudaFreeAsync(ids, s);
    cudaFreeAsync(nsel, s);
    cudaFreeAsync(tmp, s);
    CU(cudaStreamSynchronize(s));
    CU(cudaGetLastError());
    return GCGT_OK;
}

// ------------------------------------------------------------------------------------------------------------------
// C ABI
// ------------------------------------------------------------------------------------------------------------------
extern "C" void gcgt_unload(gcgt_graph* g) {
    if (!g) return;
    cudaSetDevice(g->device);
    void* bufs[] = {g->hostW ? nullptr : g->W, g->offs_alloc, g->V,      g->F,         g->N,        g->q,      g->qbits,
                    g->ctr,    g->hubq,    g->hub_ctr, g->cursor, g->fuse_ctr, g->bu_cur,   g->heavyq,   g->heavy_len, g->stats,
                    g->levels, g->parent,  g->sigma,  g->delta,     g->bc,      g->bstate,
                    g->hv_ids, g->hv_ptr,  g->hv_rem, g->hv_wptr, g->hv_bits, g->ck_prev,   g->lr_ctr, g->hv_after, g->ck_pos, g->lrq,
                    g->in_owned && !g->hostInW ? g->inW : nullptr, g->in_owned ? g->inOffs : nullptr,
                    g->crow,   g->ccol,    g->csr_hubq, g->mf,
                    g->csr_in_owned ? g->crow_in : nullptr, g->csr_in_owned ? g->ccol_in : nullptr};
    PhaseClock pc("unload");
    if (g->stream) {
        for (void* b : bufs)
            if (b) cudaFreeAsync(b, g->stream);
        cudaStreamSynchronize(g->stream);
    }
    pc.mark("free+sync");
    if (g->hostW) cudaFreeHost(g->hostW);
    if (g->hostInW) cudaFreeHost(g->hostInW);
    small_pinned_put(g->h_ctr);
    small_pinned_put(g->h_stats);
    if (g->ev0) cudaEventDestroy(g->ev0);
    if (g->ev1) cudaEventDestroy(g->ev1);
    for (auto& e : g->kevp)
        if (e) cudaEventDestroy(e);
    if (g->kev0) cudaEventDestroy(g->kev0);
    if (g->kev1) cudaEventDestroy(g->kev1);
    for (auto& e : g->sev)
        if (e) cudaEventDestroy(e);
    if (g->own_stream && g->stream) cudaStreamDestroy(g->stream);
    pc.mark("host frees+events");
    delete g;
    pc.mark("delete");
}

extern "C" gcgt_status gcgt_load(const gcgt_cgr* c, const gcgt_load_opts* opts, gcgt_graph** out) {
    gcgt_internal::clear_error();
    if (!c || !out) return fail(GCGT_EINVAL, "null argument");
    gcgt_load_opts o{};
    if (opts) o = *opts;
    if (o.nranks > 1 && (o.rank < 0 || o.rank >= o.nranks)) return fail(GCGT_EINVAL, "bad rank");
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev == 0) return fail(GCGT_ECUDA, "no CUDA device");
    if (o.device < 0 || o.device >= ndev) return fail(GCGT_EINVAL, "bad device ordinal");
    std::unique_ptr<gcgt_graph, void (*)(gcgt_graph*)> g(new gcgt_graph(), gcgt_unload);
    g->device = o.device;
    CU(cudaSetDevice(o.device));
    {   // keep freed pool memory for the next load (see galloc)
        cudaMemPool_t pool;
        if (cudaDeviceGetDefaultMemPool(&pool, o.device) == cudaSuccess) {
            uint64_t thr = UINT64_MAX;
            cudaMemPoolSetAttribute(pool, cudaMemPoolAttrReleaseThreshold, &thr);
        }
    }
    CU(cudaDeviceGetAttribute(&g->num_sms, cudaDevAttrMultiProcessorCount, o.device));
    if (o.stream) g->stream = (cudaStream_t)o.stream;
    else {
        CU(cudaStreamCreateWithFlags(&g->stream, cudaStreamNonBlocking));
        g->own_stream = true;
    }
    g->n = c->n;
    g->nbits = c->nbits;
    g->P = c->params;
    g->dir_bits = o.symmetric != 0 && !o.in_cgr;
    if (const char* tune = getenv("GCGT_TUNE")) {  // development knob: key=value,... (results never change)
        std::string t(tune);
        size_t i = 0;
        while (i < t.size()) {
            size_t j = t.find(',', i);
            if (j == std::string::npos) j = t.size();
            const std::string kv = t.substr(i, j - i);
            const size_t e = kv.find('=');
            if (e != std::string::npos) {
                const std::string k = kv.substr(0, e);
                const unsigned long v = strtoul(kv.c_str() + e + 1, nullptr, 10);
                if (k == "staged") g->staged = v != 0;
                else if (k == "persistent") g->persistent = v != 0;
                else if (k == "bu") g->bu_kernel = (uint32_t)(v == 2 ? 2 : 1);
                else if (k == "bu_words") g->bu_words = (uint32_t)std::max(1ul, std::min(8ul, v));
                else if (k == "bu_batch") g->bu_batch = (uint32_t)std::max(1ul, std::min(4ul, v));
                else if (k == "chunk") g->chunk = (uint32_t)std::max(1ul, std::min(64ul, v));
                else if (k == "nfilter") g->nfilter = (uint32_t)(v != 0);
                else if (k == "flatb") g->flatb = (uint32_t)(v != 0);
                else if (k == "fuse") g->fuse_warps = (uint32_t)std::min(8ul, v);
                else if (k == "engine") g->engine = (uint32_t)v;
                else if (k == "bu_alpha") g->bu_alpha = (uint32_t)v;
                else if (k == "bu_beta") g->bu_beta = (uint32_t)v;
                else if (k == "dir_bits") g->dir_bits = v != 0;
                else if (k == "alpha_bits") g->alpha_bits = (uint32_t)v;
                else if (k == "dir_opt") g->dir_opt_knob = v != 0;
                else if (k == "ck_c") g->ck_c = (uint32_t)std::max(1ul, v);  // 0xFFFFFFFF disables checkpoints
                else if (k == "heavy_itv") g->heavy_itv = (uint32_t)v;
                else if (k == "heavy_res") g->heavy_res = (uint32_t)v;
                else if (k == "hub_segs") g->hub_segs = (uint32_t)v;
                else if (k == "long_len") g->long_len = (uint32_t)std::max(32ul, v);
                else if (k == "wpb_max") g->wpb_max = (uint32_t)std::max(1ul, std::min(32ul, v));
            }
            i = j + 1;
        }
    }
    // 1-D vertex-range partition (§8 e): rank r owns [lo, hi), boundaries on 32-vertex words, balanced by CGR bits.
    // Records are self-contained, so the slice is a copy of whole 64-bit words plus re-based bit offsets.
    g->lo = 0;
    g->hi = c->n;
    g->nranks = o.nranks > 1 ? o.nranks : 1;
    g->rank = o.nranks > 1 ? o.rank : 0;
    if (g->nranks > 1) {
        auto bound = [&](int r) -> uint64_t {
            if (r <= 0) return 0;
            if (r >= g->nranks) return c->n;
            const uint64_t target = c->nbits / (uint64_t)g->nranks * (uint64_t)r;
            const uint64_t v = (uint64_t)(std::lower_bound(c->bit_offsets.begin(), c->bit_offsets.end(), target) -
                                          c->bit_offsets.begin());
            return std::min<uint64_t>(c->n, v & ~31ull);
        };
        g->lo = bound(g->rank);
        g->hi = std::max(g->lo, bound(g->rank + 1));
        g->dir_opt_knob = false;  // bottom-up needs the whole in-CGR: top-down only when partitioned
    }
    PhaseClock pc("load");
    g->nw = ((c->n + 31) / 32 + 1 + 3) & ~3ull;  // padded to whole 16-byte groups (commit_phase)
    const uint64_t w0 = c->bit_offsets[g->lo] / 64;
    const uint64_t nwords = (c->bit_offsets[g->hi] + 63) / 64 - w0 + 2;
    const uint64_t nloc = g->hi - g->lo;
    gcgt_status st;
    if ((o.host_resident ? (st = host_words(g.get(), &g->hostW, &g->W, c->words, w0, nwords))
                         : (st = galloc(g.get(), &g->W, nwords))) ||
        (st = galloc(g.get(), &g->offs_alloc, nloc + 1)) || (st = galloc(g.get(), &g->V, g->nw)) ||
        (st = galloc(g.get(), &g->F, g->nw)) || (st = galloc(g.get(), &g->N, g->nw)) || (st = galloc(g.get(), &g->ctr, 8)) ||
        (st = galloc(g.get(), &g->stats, 1)) || (st = galloc(g.get(), &g->levels, g->n)))
        return st;
    g->qcap = 2 * g->nw;
    if ((st = galloc(g.get(), &g->q, g->qcap))) return st;
    CU(small_pinned_get((void**)&g->h_ctr));
    CU(small_pinned_get((void**)&g->h_stats));
    CU(cudaEventCreate(&g->ev0));
    CU(cudaEventCreate(&g->ev1));
    CU(cudaEventCreate(&g->kev0));
    CU(cudaEventCreate(&g->kev1));
    for (auto& e : g->sev) CU(cudaEventCreate(&e));
    if (!o.host_resident) {
        const uint64_t avail = c->words.size() - w0;  // the host array holds >= 2 padding words
        CU(cudaMemsetAsync(g->W, 0, nwords * sizeof(uint64_t), g->stream));
        CU(cudaMemcpyAsync(g->W, c->words.data() + w0, std::min(nwords, avail) * sizeof(uint64_t),
                           cudaMemcpyHostToDevice, g->stream));
    }
    if (w0 == 0) {
        CU(cudaMemcpyAsync(g->offs_alloc, c->bit_offsets.data() + g->lo, (nloc + 1) * sizeof(uint64_t),
                           cudaMemcpyHostToDevice, g->stream));
    } else {
        std::vector<uint64_t> ro(c->bit_offsets.begin() + g->lo, c->bit_offsets.begin() + g->hi + 1);
        for (auto& x : ro) x -= w0 * 64;
        CU(cudaMemcpyAsync(g->offs_alloc, ro.data(), (nloc + 1) * sizeof(uint64_t), cudaMemcpyHostToDevice, g->stream));
        CU(cudaStreamSynchronize(g->stream));  // ro is a stack vector
    }
    pc.mark("alloc+H2D cgr", g->stream);
    g->offs = g->offs_alloc - g->lo;  // kernels index offs[u] with global vertex ids
    if (!o.host_resident) bswap_words<<<flat_grid(g.get(), nwords), kBlock, 0, g->stream>>>(g->W, nwords);
    CU(cudaMemsetAsync(g->N, 0, g->nw * 4, g->stream));
    if ((st = galloc(g.get(), &g->bstate, 8)) || (st = galloc(g.get(), &g->mf, 1))) return st;
    CU(cudaMemsetAsync(g->mf, 0, 8, g->stream));
    // in-CGR for bottom-up levels: the transpose if given, else the out-CGR itself on symmetric graphs
    if (o.in_cgr) {
        const gcgt_cgr* ic = o.in_cgr;
        if (ic->n != c->n || ic->params.zeta_k != c->params.zeta_k ||
            ic->params.min_interval_len != c->params.min_interval_len ||
            ic->params.residual_segment_len != c->params.residual_segment_len)
            return fail(GCGT_EINVAL, "in_cgr must have the same n and parameters as the CGR");
        const uint64_t inwords = (ic->nbits + 63) / 64 + 2;
        if ((o.host_resident ? (st = host_words(g.get(), &g->hostInW, &g->inW, ic->words, 0, inwords))
                             : (st = galloc(g.get(), &g->inW, inwords))) ||
            (st = galloc(g.get(), &g->inOffs, ic->n + 1)))
            return st;
        g->in_owned = true;
        if (!o.host_resident) {
            CU(cudaMemcpyAsync(g->inW, ic->words.data(), inwords * 8, cudaMemcpyHostToDevice, g->stream));
            bswap_words<<<flat_grid(g.get(), inwords), kBlock, 0, g->stream>>>(g->inW, inwords);
        }
        CU(cudaMemcpyAsync(g->inOffs, ic->bit_offsets.data(), (ic->n + 1) * 8, cudaMemcpyHostToDevice, g->stream));
        g->dir_opt = o.direction_optimizing != 0;
    } else if (o.symmetric) {
        g->inW = g->W;
        g->inOffs = g->offs;
        g->dir_opt = o.direction_optimizing != 0;
    }
    g->dir_opt = g->dir_opt && g->dir_opt_knob;
    pc.mark("in-cgr", g->stream);
    if ((st = galloc(g.get(), &g->hub_ctr, 1)) || (st = galloc(g.get(), &g->cursor, 2)) ||
        (st = galloc(g.get(), &g->fuse_ctr, 4)) || (st = galloc(g.get(), &g->bu_cur, 2)))
        return st;
    CU(cudaMemsetAsync(g->bu_cur, 0, 16, g->stream));
    CU(cudaMemsetAsync(g->cursor, 0, 16, g->stream));
    {  // epoch 1: queue entries start zeroed (epoch 0), so no stale entry can look published
        const uint32_t init[4] = {0, 0, 0, 1};
        CU(cudaMemcpyAsync(g->fuse_ctr, init, 16, cudaMemcpyHostToDevice, g->stream));
        CU(cudaStreamSynchronize(g->stream));
    }
    unsigned long long* dcount = nullptr;
    if ((st = galloc(g.get(), &dcount, 3))) return st;
    CU(cudaMemsetAsync(dcount, 0, 24, g->stream));
    {
        const int gr = flat_grid(g.get(), g->n);
        const bool seg = g->P.residual_segment_len != 0;
        cudaStream_t s = g->stream;
        switch (g->P.zeta_k) {
            case 1: seg ? count_special<1, true><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount) : count_special<1, false><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount); break;
            case 2: seg ? count_special<2, true><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount) : count_special<2, false><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount); break;
            case 3: seg ? count_special<3, true><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount) : count_special<3, false><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount); break;
            case 4: seg ? count_special<4, true><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount) : count_special<4, false><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount); break;
            default: seg ? count_special<5, true><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount) : count_special<5, false><<<gr, kBlock, 0, s>>>(g->W, g->offs, g->lo, g->hi, g->heavy_itv, g->heavy_res, g->hub_segs, g->P.min_interval_len, g->long_len, dcount); break;
        }
    }
    unsigned long long counts[3] = {0, 0, 0};
    CU(cudaMemcpyAsync(counts, dcount, 24, cudaMemcpyDeviceToHost, g->stream));
    CU(cudaStreamSynchronize(g->stream));
    cudaFreeAsync(dcount, g->stream);
    pc.mark("count_special");
    const uint64_t nhubs = counts[0], nheavy = counts[1], nlong = counts[2];
    if ((st = galloc(g.get(), &g->heavyq, nheavy + 1)) || (st = galloc(g.get(), &g->heavy_len, 1))) return st;
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, g->stream));
    if ((st = galloc(g.get(), &g->hubq, nhubs + nheavy + 1))) return st;
    CU(cudaMemsetAsync(g->hubq, 0, (nhubs + nheavy + 1) * sizeof(HubEntry), g->stream));
    if ((st = build_checkpoints(g.get()))) return st;
    pc.mark("checkpoints", g->stream);
    if ((st = galloc(g.get(), &g->lrq, nlong + 1))) return st;
    CU(cudaMemsetAsync(g->lrq, 0, (nlong + 1) * sizeof(LongRange), g->stream));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 8, g->stream));
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
    pc.mark("end");
    *out = g.release();
    return GCGT_OK;
}


// Uncompressed baseline load (§8 f3): plain CSR on the device; in-lists = the host transpose (counting sort) or the
// CSR itself when symmetric.  Shares the frontier buffers and counters with the CGR path.
extern "C" gcgt_status gcgt_load_csr(const gcgt_csr* csr, const gcgt_load_opts* opts, gcgt_graph** out) {
    gcgt_internal::clear_error();
    if (!csr || !out || (csr->n && !csr->row_offsets)) return fail(GCGT_EINVAL, "null argument");
    gcgt_load_opts o{};
    if (opts) o = *opts;
    if (o.nranks > 1) return fail(GCGT_EINVAL, "CSR baseline: single GPU only");
    const uint64_t n = csr->n, m = n ? csr->row_offsets[n] : 0;
    if (n >= 0xFFFFFFFFull) return fail(GCGT_ERANGE, "n must fit 32-bit ids");
    if (m && !csr->cols) return fail(GCGT_EINVAL, "null cols");
    for (uint64_t v = 0; v < n; v++)
        if (csr->row_offsets[v + 1] < csr->row_offsets[v]) return fail(GCGT_EINVAL, "row_offsets not monotone");
    for (uint64_t e = 0; e < m; e++)
        if (csr->cols[e] >= n) return fail(GCGT_ERANGE, "column id >= n");
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev == 0) return fail(GCGT_ECUDA, "no CUDA device");
    if (o.device < 0 || o.device >= ndev) return fail(GCGT_EINVAL, "bad device ordinal");
    std::unique_ptr<gcgt_graph, void (*)(gcgt_graph*)> g(new gcgt_graph(), gcgt_unload);
    g->device = o.device;
    g->is_csr = true;
    CU(cudaSetDevice(o.device));
    CU(cudaDeviceGetAttribute(&g->num_sms, cudaDevAttrMultiProcessorCount, o.device));
    if (o.stream) g->stream = (cudaStream_t)o.stream;
    else {
        CU(cudaStreamCreateWithFlags(&g->stream, cudaStreamNonBlocking));
        g->own_stream = true;
    }
    g->dir_bits = o.symmetric != 0;
    if (const char* tune = getenv("GCGT_TUNE")) {  // the direction-switch knobs apply here too
        std::string t(tune);
        for (const char* k : {"bu_alpha=", "bu_beta=", "alpha_bits=", "dir_bits="}) {
            const size_t i = t.find(k);
            if (i != std::string::npos && (i == 0 || t[i - 1] == ',')) {
                const uint32_t v = (uint32_t)strtoul(t.c_str() + i + strlen(k), nullptr, 10);
                if (k[0] == 'b' && k[3] == 'a') g->bu_alpha = v;
                else if (k[0] == 'b') g->bu_beta = v;
                else if (k[0] == 'a') g->alpha_bits = v;
                else g->dir_bits = v != 0;
            }
        }
    }
    g->n = n;
    g->lo = 0;
    g->hi = n;
    g->nw = ((n + 31) / 32 + 1 + 3) & ~3ull;
    cudaStream_t s = g->stream;
    gcgt_status st;
    if ((st = galloc(g.get(), &g->crow, n + 1)) || (st = galloc(g.get(), &g->ccol, m)) ||
        (st = galloc(g.get(), &g->V, g->nw)) || (st = galloc(g.get(), &g->F, g->nw)) ||
        (st = galloc(g.get(), &g->N, g->nw)) || (st = galloc(g.get(), &g->ctr, 8)) ||
        (st = galloc(g.get(), &g->stats, 1)) || (st = galloc(g.get(), &g->levels, n)) ||
        (st = galloc(g.get(), &g->bstate, 8)) || (st = galloc(g.get(), &g->hub_ctr, 1)) ||
        (st = galloc(g.get(), &g->mf, 1)) ||
        (st = galloc(g.get(), &g->cursor, 2)))
        return st;
    g->qcap = 2 * g->nw;
    if ((st = galloc(g.get(), &g->q, g->qcap))) return st;
    CU(small_pinned_get((void**)&g->h_ctr));
    CU(small_pinned_get((void**)&g->h_stats));
    CU(cudaEventCreate(&g->ev0));
    CU(cudaEventCreate(&g->ev1));
    CU(cudaEventCreate(&g->kev0));
    CU(cudaEventCreate(&g->kev1));
    for (auto& e : g->sev) CU(cudaEventCreate(&e));
    CU(cudaMemcpyAsync(g->crow, csr->row_offsets, (n + 1) * 8, cudaMemcpyHostToDevice, s));
    if (m) CU(cudaMemcpyAsync(g->ccol, csr->cols, m * 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemsetAsync(g->N, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->cursor, 0, 16, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->mf, 0, 8, s));
    g->nbits = m;  // the CSR's "record bits" for the direction test: arcs
    uint64_t nhub = 0;
    for (uint64_t v = 0; v < n; v++) nhub += csr->row_offsets[v + 1] - csr->row_offsets[v] > kCsrHub;
    CsrHubEntry* hubq = nullptr;
    if ((st = galloc(g.get(), &hubq, nhub + 1))) return st;
    g->csr_hubq = hubq;
    if (o.direction_optimizing) {
        if (o.symmetric) {
            g->crow_in = g->crow;
            g->ccol_in = g->ccol;
            g->dir_opt = true;
        } else {
            std::vector<uint64_t> tro(n + 1, 0);
            std::vector<uint32_t> tco(m);
            for (uint64_t e = 0; e < m; e++) tro[csr->cols[e] + 1]++;
            for (uint64_t v = 0; v < n; v++) tro[v + 1] += tro[v];
            std::vector<uint64_t> pos(tro.begin(), tro.end() - 1);
            for (uint64_t u = 0; u < n; u++)
                for (uint64_t e = csr->row_offsets[u]; e < csr->row_offsets[u + 1]; e++)
                    tco[pos[csr->cols[e]]++] = (uint32_t)u;
            if ((st = galloc(g.get(), &g->crow_in, n + 1)) || (st = galloc(g.get(), &g->ccol_in, m))) return st;
            g->csr_in_owned = true;
            CU(cudaMemcpyAsync(g->crow_in, tro.data(), (n + 1) * 8, cudaMemcpyHostToDevice, s));
            if (m) CU(cudaMemcpyAsync(g->ccol_in, tco.data(), m * 4, cudaMemcpyHostToDevice, s));
            CU(cudaStreamSynchronize(s));  // tro / tco are host vectors
            g->dir_opt = true;
        }
    }
    CU(cudaStreamSynchronize(s));
    CU(cudaGetLastError());
    *out = g.release();
    return GCGT_OK;
}

// ---- test hook: the warp decoder on a caller bit array (Fig. 5 pin) --------------------------------------------------
namespace {
template <int K, int WIN>
__global__ void debug_warp_decode_kernel(const uint64_t* W, uint64_t count, uint64_t* vals, uint32_t* tpos,
                                         uint32_t* tflags, uint32_t* rounds) {
    uint64_t v;
    uint32_t len;
    window_step<K, WIN, true>(W, 0, v, len, tpos, tflags, rounds);
    warp_decode<K>(W, 0, count, [&](uint64_t, uint32_t, uint64_t idx, uint64_t val, bool act) {
        if (act) vals[idx] = val;
    });
}

template <int K>
void launch_debug(uint32_t win, const uint64_t* W, uint64_t count, uint64_t* vals, uint32_t* tp, uint32_t* tf,
                  uint32_t* r) {
    if (win == 16) debug_warp_decode_kernel<K, 16><<<1, 32>>>(W, count, vals, tp, tf, r);
    else debug_warp_decode_kernel<K, 32><<<1, 32>>>(W, count, vals, tp, tf, r);
}
}  // namespace

extern "C" gcgt_status gcgt_debug_warp_decode(const uint8_t* bytes, uint64_t nbits, uint32_t zeta_k, uint32_t window,
                                              uint64_t count, uint64_t* vals, uint32_t* trace_pos,
                                              uint32_t* trace_flags, uint32_t* rounds) {
    gcgt_internal::clear_error();
    if (!bytes || !vals || !trace_pos || !trace_flags || !rounds) return fail(GCGT_EINVAL, "null argument");
    if (zeta_k < 1 || zeta_k > 5 || (window != 16 && window != 32)) return fail(GCGT_EINVAL, "bad zeta_k / window");
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev == 0) return fail(GCGT_ECUDA, "no CUDA device");
    const uint64_t nwords = (nbits + 63) / 64 + 4;
    std::vector<uint64_t> h(nwords, 0);
    memcpy(h.data(), bytes, (nbits + 7) / 8);
    for (auto& x : h) x = __builtin_bswap64(x);
    uint64_t *dW = nullptr, *dv = nullptr;
    uint32_t *dp = nullptr, *df = nullptr, *dr = nullptr;
    gcgt_status st = GCGT_OK;
    if ((st = dalloc(&dW, nwords)) || (st = dalloc(&dv, count + 1)) || (st = dalloc(&dp, 6 * 32)) ||
        (st = dalloc(&df, 6 * 32)) || (st = dalloc(&dr, 1))) {
        cudaFree(dW); cudaFree(dv); cudaFree(dp); cudaFree(df); cudaFree(dr);
        return st;
    }
    cudaMemcpy(dW, h.data(), nwords * 8, cudaMemcpyHostToDevice);
    cudaMemset(dp, 0xff, 6 * 32 * 4);
    cudaMemset(df, 0, 6 * 32 * 4);
    switch (zeta_k) {
        case 1: launch_debug<1>(window, dW, count, dv, dp, df, dr); break;
        case 2: launch_debug<2>(window, dW, count, dv, dp, df, dr); break;
        case 3: launch_debug<3>(window, dW, count, dv, dp, df, dr); break;
        case 4: launch_debug<4>(window, dW, count, dv, dp, df, dr); break;
        default: launch_debug<5>(window, dW, count, dv, dp, df, dr); break;
    }
    cudaError_t e = cudaDeviceSynchronize();
    if (e == cudaSuccess) {
        cudaMemcpy(vals, dv, count * 8, cudaMemcpyDeviceToHost);
        cudaMemcpy(trace_pos, dp, 6 * 32 * 4, cudaMemcpyDeviceToHost);
        cudaMemcpy(trace_flags, df, 6 * 32 * 4, cudaMemcpyDeviceToHost);
        e = cudaMemcpy(rounds, dr, 4, cudaMemcpyDeviceToHost);
    }
    cudaFree(dW); cudaFree(dv); cudaFree(dp); cudaFree(df); cudaFree(dr);
    if (e != cudaSuccess) return fail(GCGT_ECUDA, cudaGetErrorString(e));
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_profile(gcgt_graph* g, int enable) {
    if (!g) return fail(GCGT_EINVAL, "null graph");
    g->profile = enable != 0;
    g->spans = enable >= 2;
    g->kev_n = 0;
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_profile_spans(const gcgt_graph* g, double* ms, int count) {
    if (!g || !ms) return fail(GCGT_EINVAL, "null argument");
    for (int k = 0; k < count && k < 4; k++) ms[k] = g->span_ms[k];
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_graph_range(const gcgt_graph* g, uint64_t* lo, uint64_t* hi) {
    if (!g) return fail(GCGT_EINVAL, "null graph");
    if (lo) *lo = g->lo;
    if (hi) *hi = g->hi;
    return GCGT_OK;
}


// ---- uncompressed-CSR baseline (§8 f3, csr_bfs.cuh) -------------------------------------------------------------
gcgt_status csr_bfs(gcgt_graph* g, uint32_t source, int32_t* levels, int placement, gcgt_stats* stats) {
    cudaStream_t s = g->stream;
    CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->F, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
    CU(cudaMemsetAsync(g->ctr, 0, 8 * 4, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, sizeof(unsigned long long), s));
    uint32_t* q[2] = {g->q, g->q + g->nw};
    bfs_seed<<<1, 1, 0, s>>>(source, g->V, g->F, q[0], g->ctr + 0, nullptr, g->levels, g->bstate);
    g->launches = 1;
    static int per_sm = 0;
    if (!per_sm) {
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, csr_expand_kernel<QueueFront>, kBlock, 0);
        if (per_sm < 1) per_sm = 1;
    }
    static int per_sm_bu = 0;
    if (!per_sm_bu) {
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm_bu, csr_bu_kernel, kBlock, 0);
        if (per_sm_bu < 1) per_sm_bu = 1;
    }
    const int egrid = per_sm * g->num_sms;
    const int bgrid = (int)std::max<uint64_t>(1, std::min<uint64_t>((g->nw + kWarps - 1) / kWarps,
                                                                    (uint64_t)per_sm_bu * g->num_sms));
    CsrHubEntry* hubq = (CsrHubEntry*)g->csr_hubq;
    uint64_t qlen = 1;
    uint32_t level = 0;
    gcgt_status st;
    while (qlen) {
        const uint32_t nlev = g->spans ? 1 : std::min<uint32_t>(g->chunk, gcgt_graph::kKev);
        for (uint32_t i = 0; i < nlev; i++, level++) {
            const int cur = level & 1, nxt = cur ^ 1;
            const QueueFront fr{q[cur], g->ctr + cur, g->F, nullptr};
            const BfsApp app{g->V, g->N, g->levels, (int32_t)level, g->nfilter};
            if ((st = kprof_begin(g))) return st;
            if (g->spans) CU(cudaEventRecord(g->sev[0], s));
            csr_expand_kernel<QueueFront><<<egrid, kBlock, 0, s>>>(g->crow, g->ccol, fr, app, g->cursor, hubq,
                                                                    g->hub_ctr, g->dir_opt ? g->bstate : nullptr,
                                                                    g->stats);
            if (g->spans) CU(cudaEventRecord(g->sev[1], s));
            csr_hub_kernel<<<hub_grid(g), kBlock, 0, s>>>(g->ccol, hubq, g->hub_ctr, app, g->stats);
            if (g->spans) CU(cudaEventRecord(g->sev[2], s));
            if (g->dir_opt)
                csr_bu_kernel<<<bgrid, kBlock, 0, s>>>(g->crow_in, g->ccol_in, g->V, g->F, g->N, g->n, g->bstate,
                                                        g->stats);
            if (g->spans) CU(cudaEventRecord(g->sev[3], s));
            if ((st = kprof_end(g))) return st;
            commit_dense<<<flat_grid(g, g->nw), kBlock, 0, s>>>(g->V, g->F, g->N, 0, g->nw, q[nxt], g->ctr + nxt,
                                                                 nullptr, g->ctr + cur, g->hub_ctr, nullptr,
                                                                 g->levels, (int32_t)level + 1, g->bstate + 2,
                                                                 nullptr, g->dir_bits && g->dir_opt ? g->crow : nullptr,
                                                                 g->dir_bits && g->dir_opt ? g->mf : nullptr,
                DecideArgs{g->bstate, g->n, g->bu_alpha, g->bu_beta, g->dir_opt ? 1 : 0, g->ctr + nxt, g->ctr + 6,
                           g->dir_bits && g->dir_opt ? g->mf : nullptr,
                           (double)g->nbits / (double)std::max<uint64_t>(1, g->n), g->alpha_bits, g->ctr + 7});
            g->launches += 3 + (g->dir_opt ? 1 : 0);
            if (g->spans) {
                CU(cudaEventRecord(g->sev[4], s));
                CU(cudaEventSynchronize(g->sev[4]));
                for (int k = 0; k < 4; k++) {
                    float ms = 0;
                    CU(cudaEventElapsedTime(&ms, g->sev[k], g->sev[k + 1]));
                    g->span_ms[k] += ms;
                }
            }
        }
        CU(cudaMemcpyAsync(g->h_ctr + 6, g->ctr + 6, 4, cudaMemcpyDeviceToHost, s));
        CU(cudaMemcpyAsync(g->h_ctr + (level & 1), g->ctr + (level & 1), 4, cudaMemcpyDeviceToHost, s));
        CU(cudaStreamSynchronize(s));
        if ((st = kprof_collect(g))) return st;
        qlen = g->h_ctr[level & 1];
    }
    if ((st = copy_out(g, levels, g->levels, g->n * 4, placement))) return st;
    return end_call(g, stats, g->h_ctr[6] + 1);
}

extern "C" gcgt_status gcgt_bfs(gcgt_graph* g, uint32_t source, int32_t* levels, int placement, gcgt_stats* stats) {
    if (!g || !levels) return fail(GCGT_EINVAL, "null argument");
    if (g->nranks > 1) return fail(GCGT_EINVAL, "partitioned graph: use the gcgt_dist_* steps (dist.py)");
    if (source >= g->n) return fail(GCGT_ERANGE, "source >= n");
    gcgt_status st;
    if ((st = begin_call(g))) return st;
    if (g->is_csr) return csr_bfs(g, source, levels, placement, stats);
    cudaStream_t s = g->stream;
    CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->F, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
    CU(cudaMemsetAsync(g->ctr, 0, 8 * 4, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, sizeof(unsigned long long), s));
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
    uint32_t* q[2] = {g->q, g->q + g->nw};
    bfs_seed<<<1, 1, 0, s>>>(source, g->V, g->F, q[0], g->ctr + 0, nullptr, g->levels, g->bstate);
    g->launches = 1;
    Ctx c = make_ctx(g);
    if (g->dir_opt) c.dir = g->bstate;
    uint64_t qlen = 1;
    uint32_t level = 0;
    if (g->persistent) {
        const BfsPersist b{q[0], q[1], g->ctr, g->V, g->F, g->N, g->levels, g->nw, g->wpb_max};
        if ((st = kprof_begin(g))) return st;
        const cudaError_t e = launch_bfs_persistent(g, s, c, b);
        if (e == cudaSuccess) {
            g->launches += 1;
            if ((st = kprof_end(g))) return st;
            CU(cudaMemcpyAsync(g->h_ctr + 6, g->ctr + 6, 4, cudaMemcpyDeviceToHost, s));
            CU(cudaStreamSynchronize(s));
            if ((st = kprof_collect(g))) return st;
            level = g->h_ctr[6];
            qlen = 0;  // done
        } else {
            cudaGetLastError();  // cannot co-schedule: fall through to the host-driven loop
            g->persistent = false;
        }
    }
    // Host-driven level loop without a per-level wait: the kernels size their work from the device-resident queue
    // length, so the host enqueues kChunk levels at a time and checks for an empty queue once per chunk (levels
    // enqueued past the end find an empty queue and exit at once).  With profiling on, the loop waits per level to
    // time the expansion kernel.
    while (qlen) {
        const uint32_t nlev = g->spans ? 1 : std::min<uint32_t>(g->chunk, gcgt_graph::kKev);
        for (uint32_t i = 0; i < nlev; i++, level++) {
            const int cur = level & 1, nxt = cur ^ 1;
            int grid;
            uint32_t wpb;
            frontier_launch(g, level == 0 ? 1 : (uint64_t)g->nw, &grid, &wpb);
            if (level == 0) wpb = 1;
            else wpb = 0;  // device-side sizing
            const QueueFront fr{q[cur], g->ctr + cur, g->F, nullptr};
            const BfsApp app{g->V, g->N, g->levels, (int32_t)level, g->nfilter};
            // profiled span = the level's expansion: top-down kernel (+ heavy pass + hub segments) or bottom-up
            if ((st = kprof_begin(g))) return st;
            if (g->spans) CU(cudaEventRecord(g->sev[0], s));
            launch_expand(g->P, g->staged, grid, s, c, fr, app, wpb);
            launch_heavy(g, s, c, app);
            if (g->spans) CU(cudaEventRecord(g->sev[1], s));
            launch_hub(g->P, g->staged, hub_grid(g), s, c, app);
            if (g->spans) CU(cudaEventRecord(g->sev[2], s));
            if (g->dir_opt) launch_bu(g, s);
            if (g->spans) CU(cudaEventRecord(g->sev[3], s));
            if ((st = kprof_end(g))) return st;
            commit_dense<<<flat_grid(g, g->nw), kBlock, 0, s>>>(g->V, g->F, g->N, 0, g->nw, q[nxt], g->ctr + nxt,
                                                                 nullptr, g->ctr + cur, g->hub_ctr, g->heavy_len,
                                                                 g->levels, (int32_t)level + 1, g->bstate + 2,
                                                                 g->lr_ctr, g->dir_bits && g->dir_opt ? g->offs : nullptr,
                                                                 g->dir_bits && g->dir_opt ? g->mf : nullptr,
                DecideArgs{g->bstate, g->n, g->bu_alpha, g->bu_beta, g->dir_opt ? 1 : 0, g->ctr + nxt, g->ctr + 6,
                           g->dir_bits && g->dir_opt ? g->mf : nullptr,
                           (double)g->nbits / (double)std::max<uint64_t>(1, g->n), g->alpha_bits, g->ctr + 7});
            if (g->spans) {  // span profiling waits per level (nlev = 1)
                CU(cudaEventRecord(g->sev[4], s));
                CU(cudaEventSynchronize(g->sev[4]));
                float lms[4];
                for (int k = 0; k < 4; k++) {
                    CU(cudaEventElapsedTime(&lms[k], g->sev[k], g->sev[k + 1]));
                    g->span_ms[k] += lms[k];
                }
                if (getenv("GCGT_TRACE")) {  // development aid (tools/trace_bfs.py): one line per level on stderr
                    uint32_t hb[4], hq = 0;
                    CU(cudaMemcpy(hb, g->bstate, 16, cudaMemcpyDeviceToHost));
                    CU(cudaMemcpy(&hq, g->ctr + nxt, 4, cudaMemcpyDeviceToHost));
                    fprintf(stderr, "level %3u next_dir %u visited %10u new %9u next_words %8u | exp %.4f hub %.4f "
                            "bu %.4f commit %.4f ms\n", level, hb[0], hb[1], hb[3], hq, lms[0], lms[1], lms[2], lms[3]);
                }
            }
            g->launches += 2 + (g->P.residual_segment_len ? 1 : 0) + (g->dir_opt ? 1 : 0) + (heavy_active(g) ? 1 : 0);
        }
        CU(cudaMemcpyAsync(g->h_ctr + 6, g->ctr + 6, 4, cudaMemcpyDeviceToHost, s));
        CU(cudaMemcpyAsync(g->h_ctr + (level & 1), g->ctr + (level & 1), 4, cudaMemcpyDeviceToHost, s));
        CU(cudaStreamSynchronize(s));
        if ((st = kprof_collect(g))) return st;
        qlen = g->h_ctr[level & 1];
    }
    if (!g->persistent || level == 0) level = g->h_ctr[6] + 1;  // non-empty levels expanded (seed level included)
    if ((st = copy_out(g, levels, g->levels, g->n * 4, placement))) return st;
    return end_call(g, stats, level);
}

extern "C" gcgt_status gcgt_cc(gcgt_graph* g, uint32_t* labels, int placement, gcgt_stats* stats) {
    if (!g || !labels) return fail(GCGT_EINVAL, "null argument");
    if (g->is_csr) return fail(GCGT_EINVAL, "CSR baseline graph: BFS only");
    if (g->nranks > 1) return fail(GCGT_EINVAL, "partitioned graph: use the gcgt_dist_* steps (dist.py)");
    gcgt_status st;
    if (!g->parent && (st = galloc(g, &g->parent, g->n))) return st;
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    CU(cudaMemsetAsync(g->hub_ctr, 0, sizeof(unsigned long long), s));
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
    cc_init<<<flat_grid(g, g->n), kBlock, 0, s>>>(g->parent, g->n);
    const Ctx c = make_ctx(g);
    const DenseFront fr{g->lo, g->hi};
    const CcApp app{g->parent, 0, nullptr, 0};
    int grid;
    uint32_t wpb;
    frontier_launch(g, (g->hi - g->lo + 31) / 32 + 1, &grid, &wpb);
    if ((st = kprof_begin(g))) return st;
    launch_expand(g->P, g->staged, grid, s, c, fr, app, wpb);
    if ((st = kprof_end(g))) return st;
    launch_heavy(g, s, c, app);
    launch_hub(g->P, g->staged, hub_grid(g), s, c, app);
    cc_jump<<<flat_grid(g, g->n), kBlock, 0, s>>>(g->parent, g->n);
    if ((st = copy_out(g, labels, g->parent, g->n * 4, placement))) return st;
    CU(cudaStreamSynchronize(s));
    if ((st = kprof_collect(g))) return st;
    return end_call(g, stats, 1);
}

extern "C" gcgt_status gcgt_bc(gcgt_graph* g, const uint32_t* sources, uint32_t k, double* bc, int placement,
                               gcgt_stats* stats) {
    if (g && g->is_csr) return fail(GCGT_EINVAL, "CSR baseline graph: BFS only");
    if (!g || !bc || (k && !sources)) return fail(GCGT_EINVAL, "null argument");
    if (g->nranks > 1) return fail(GCGT_EINVAL, "partitioned graph: BC shards sources over full replicas (dist.py)");
    for (uint32_t i = 0; i < k; i++)
        if (sources[i] >= g->n) return fail(GCGT_ERANGE, "source >= n");
    gcgt_status st;
    if (!g->sigma) {
        if ((st = galloc(g, &g->sigma, g->n)) || (st = galloc(g, &g->delta, g->n)) || (st = galloc(g, &g->bc, g->n)) ||
            (st = galloc(g, &g->qbits, g->n + g->nw)))
            return st;
        uint32_t* bigq = nullptr;
        if ((st = galloc(g, &bigq, g->n + g->nw))) return st;
        cudaFreeAsync(g->q, g->stream);
        g->q = bigq;
        g->qcap = g->n + g->nw;
    }
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    const Ctx c = make_ctx(g);
    CU(cudaMemsetAsync(g->bc, 0, g->n * 8, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, sizeof(unsigned long long), s));
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
    std::vector<uint32_t> lvl_off;
    for (uint32_t si = 0; si < k; si++) {
        const uint32_t src = sources[si];
        CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
        CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
        CU(cudaMemsetAsync(g->sigma, 0, g->n * 8, s));
        CU(cudaMemsetAsync(g->delta, 0, g->n * 8, s));
        CU(cudaMemsetAsync(g->ctr, 0, 8 * 4, s));
        const double one = 1.0;
        CU(cudaMemcpyAsync(g->sigma + src, &one, 8, cudaMemcpyHostToDevice, s));
        // level d occupies q[lvl_off[d] .. lvl_off[d+1]) (words) with qbits (their frontier bits)
        bfs_seed<<<1, 1, 0, s>>>(src, g->V, nullptr, g->q, g->ctr + 2, g->qbits);
        lvl_off.assign(1, 0);
        uint32_t total = 1, level = 0;
        for (;;) {
            const uint32_t off = lvl_off.back(), qlen = total - off;
            lvl_off.push_back(total);
            if (!qlen) break;
            int grid;
            uint32_t wpb;
            frontier_launch(g, qlen, &grid, &wpb);
            // ctr[2] holds this level's length (seed or the previous commit), ctr[3] receives the next one
            const QueueFront fr{g->q + off, g->ctr + 2 + (level & 1), nullptr, g->qbits + off};
            const BcFwdApp app{g->V, g->N, g->levels, g->sigma, (int32_t)level, 0.0};
            if ((st = kprof_begin(g))) return st;
            launch_expand(g->P, g->staged, grid, s, c, fr, app, wpb);
            if ((st = kprof_end(g))) return st;
            launch_heavy(g, s, c, app);
            launch_hub(g->P, g->staged, hub_grid(g), s, c, app);
            commit_dense<<<flat_grid(g, g->nw), kBlock, 0, s>>>(g->V, nullptr, g->N, 0, g->nw, g->q + total,
                                                                 g->ctr + 2 + ((level + 1) & 1), g->qbits + total,
                                                                 g->ctr + 2 + (level & 1), g->hub_ctr,
                                                                 g->heavy_len, nullptr, 0, nullptr, g->lr_ctr);
            CU(cudaMemcpyAsync(g->h_ctr + 1, g->ctr + 2 + ((level + 1) & 1), 4, cudaMemcpyDeviceToHost, s));
            CU(cudaStreamSynchronize(s));
            if ((st = kprof_collect(g))) return st;
            total += g->h_ctr[1];
            level++;
        }
        const int D = (int)lvl_off.size() - 2;  // levels 0..D-1
        for (int d = D - 1; d >= 0; d--) {
            const uint32_t off = lvl_off[d], qlen = lvl_off[d + 1] - off;
            CU(cudaMemcpyAsync(g->ctr + 4, &qlen, 4, cudaMemcpyHostToDevice, s));
            int grid;
            uint32_t wpb;
            frontier_launch(g, qlen, &grid, &wpb);
            const QueueFront fr{g->q + off, g->ctr + 4, nullptr, g->qbits + off};
            const BcBwdApp app{g->levels, g->sigma, g->delta, g->bc, d + 1, src, 0, 0.0, 0.0};
            launch_expand(g->P, g->staged, grid, s, c, fr, app, wpb);
            launch_heavy(g, s, c, app);
            launch_hub(g->P, g->staged, hub_grid(g), s, c, app);
            CU(cudaMemsetAsync(g->hub_ctr, 0, sizeof(unsigned long long), s));
            CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
            CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
        }
    }
    if ((st = copy_out(g, bc, g->bc, g->n * 8, placement))) return st;
    return end_call(g, stats, k);
}

// ------------------------------------------------------------------------------------------------------------------
// Partitioned (multi-GPU) steps.  The caller (paper_conf_sigmod_shalt19_b200/dist.py) runs the collectives between
// them; all bitmaps crossing the boundary are device arrays of ceil(n/32) 32-bit words (bit v%32 of word v/32).
// ------------------------------------------------------------------------------------------------------------------
namespace {
gcgt_status dist_sync(gcgt_graph* g) {
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
    return GCGT_OK;
}
}  // namespace

extern "C" gcgt_status gcgt_dist_bfs_begin(gcgt_graph* g, uint32_t source) {
    gcgt_internal::clear_error();
    if (!g) return fail(GCGT_EINVAL, "null graph");
    if (g->is_csr) return fail(GCGT_EINVAL, "CSR baseline graph: single-GPU BFS only");
    if (source >= g->n) return fail(GCGT_ERANGE, "source >= n");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->F, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
    CU(cudaMemsetAsync(g->ctr, 0, 8 * 4, s));
    bfs_seed<<<1, 1, 0, s>>>(source, g->V, g->F, g->q, g->ctr, nullptr, g->levels, nullptr);
    return dist_sync(g);
}

extern "C" gcgt_status gcgt_dist_bfs_expand(gcgt_graph* g, uint32_t level, uint32_t* cand) {
    gcgt_internal::clear_error();
    if (!g || !cand) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    CU(cudaMemsetAsync(cand, 0, ((g->n + 31) / 32) * 4, s));
    const Ctx c = make_ctx(g);
    const BitsFront fr{g->F, g->lo, g->hi};
    const BfsApp app{g->V, cand, g->levels, (int32_t)level};
    int grid;
    uint32_t wpb;
    frontier_launch(g, (g->hi - g->lo + 31) / 32 + 1, &grid, &wpb);
    launch_expand(g->P, g->staged, grid, s, c, fr, app, 0);
    launch_heavy(g, s, c, app);
    launch_hub(g->P, g->staged, hub_grid(g), s, c, app);
    CU(cudaMemsetAsync(g->hub_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
    return dist_sync(g);
}

extern "C" gcgt_status gcgt_dist_bfs_commit(gcgt_graph* g, uint32_t level, const uint32_t* recv, uint32_t nparts,
                                            uint32_t* fslice, uint64_t* new_count) {
    gcgt_internal::clear_error();
    if (!g || !recv || !fslice || !new_count || nparts == 0) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    const uint64_t w_lo = g->lo / 32, nlw = (g->hi + 31) / 32 - w_lo;
    unsigned long long* cnt = (unsigned long long*)g->stats;  // scratch: reuse the stats block
    CU(cudaMemsetAsync(cnt, 0, 8, s));
    if (nlw)
        dist_commit<<<flat_grid(g, nlw * 32), kBlock, 0, s>>>(recv, nparts, w_lo, nlw, g->V, fslice, g->levels,
                                                               (int32_t)level + 1, g->n, cnt);
    CU(cudaMemcpyAsync(g->h_stats, cnt, 8, cudaMemcpyDeviceToHost, s));
    gcgt_status st = dist_sync(g);
    if (st) return st;
    *new_count = g->h_stats->vertices;
    CU(cudaMemsetAsync(g->stats, 0, sizeof(Stats), s));
    return dist_sync(g);
}

extern "C" gcgt_status gcgt_dist_bfs_absorb(gcgt_graph* g, const uint32_t* frontier) {
    gcgt_internal::clear_error();
    if (!g || !frontier) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    const uint64_t nwf = (g->n + 31) / 32;
    dist_absorb<<<flat_grid(g, nwf), kBlock, 0, g->stream>>>(frontier, g->F, g->V, nwf);
    return dist_sync(g);
}

extern "C" gcgt_status gcgt_dist_bfs_levels(gcgt_graph* g, int32_t* levels_owned, int placement) {
    gcgt_internal::clear_error();
    if (!g || !levels_owned) return fail(GCGT_EINVAL, "null argument");
    gcgt_status st;
    if ((st = copy_out(g, levels_owned, g->levels + g->lo, (g->hi - g->lo) * 4, placement))) return st;
    return dist_sync(g);
}

extern "C" gcgt_status gcgt_dist_cc_hook(gcgt_graph* g, uint32_t* parent, uint64_t* hooks) {
    gcgt_internal::clear_error();
    if (!g || !parent || !hooks) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    uint32_t* hc = g->ctr + 7;
    CU(cudaMemsetAsync(hc, 0, 4, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->lr_ctr, 0, 8, s));
    CU(cudaMemsetAsync(g->heavy_len, 0, 4, s));
    const Ctx c = make_ctx(g);
    const DenseFront fr{g->lo, g->hi};
    const CcApp app{parent, 0, hc, 0};
    int grid;
    uint32_t wpb;
    frontier_launch(g, (g->hi - g->lo + 31) / 32 + 1, &grid, &wpb);
    launch_expand(g->P, g->staged, grid, s, c, fr, app, wpb);
    launch_heavy(g, s, c, app);
    launch_hub(g->P, g->staged, hub_grid(g), s, c, app);
    CU(cudaMemcpyAsync(g->h_ctr + 7, hc, 4, cudaMemcpyDeviceToHost, s));
    gcgt_status st = dist_sync(g);
    if (st) return st;
    *hooks = g->h_ctr[7];
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_cc_jump(gcgt_graph* g, uint32_t* parent) {
    gcgt_internal::clear_error();
    if (!g || !parent) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cc_jump<<<flat_grid(g, g->n), kBlock, 0, g->stream>>>(parent, g->n);
    return dist_sync(g);
}

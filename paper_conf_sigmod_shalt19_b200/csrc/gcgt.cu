// gcgt.cu — B200 (sm_100a) device path of GCGT: device residency of the CGR, the level loops of BFS / CC / BC, the
// partitioned (multi-GPU) steps, and the C ABI around them (include/gcgt.h).
//
// Pipeline per level (expansion - filtering - contraction, §6, Fig. 7(a)):
//   top-down   expand_kernel (records staged through shared memory, lane per vertex for the header and intervals,
//              residual segments through a per-warp pool drained by a flat lane-refill loop) and hub_kernel
//              (long interval areas and multi-segment vertices over the whole grid)        — expand.cuh
//   bottom-up  bu_kernel (in-records scanned until the first frontier parent)                — bottomup.cuh
//   contract   commit_kernel (N -> V / F / levels / next queue; direction; level counter)   — contract.cuh
// The level state lives on the device, so BFS runs as one CUDA graph: a while-node whose body holds two levels,
// each an if/else node choosing top-down or bottom-up from the direction the previous contraction decided.  No host
// round trip and no empty grid per level.
#include <cuda_runtime.h>
#include <stdio.h>
#include <string.h>

#include <algorithm>
#include <chrono>
#include <memory>
#include <mutex>
#include <string>
#include <vector>

#include "bottomup.cuh"
#include "contract.cuh"
#include "csr_bfs.cuh"
#include "expand.cuh"
#include "internal.h"

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
extern "C" const char* gcgt_version(void) { return "gcgt-b200 0.2 (sm_100a)"; }

#define CU(call)                                                                                          \
    do {                                                                                                  \
        cudaError_t e_ = (call);                                                                          \
        if (e_ != cudaSuccess) return fail(GCGT_ECUDA, std::string(#call) + ": " + cudaGetErrorString(e_)); \
    } while (0)

// ------------------------------------------------------------------------------------------------------------------
// device graph
// ------------------------------------------------------------------------------------------------------------------
// A CGR (or the in-CGR) resident on the device: stream words of the owned records and their bit offsets.
struct DevCgr {
    uint64_t* W = nullptr;      // device words (or the device alias of hostW)
    uint64_t* hostW = nullptr;  // host-resident CGR (§8 f4): pinned, mapped host words
    uint64_t* anc = nullptr;    // compact offsets: u64 anchor per 256 vertices
    uint32_t* rel = nullptr;    //                  u32 offset relative to the anchor
    uint64_t* full = nullptr;   // plain u64 offsets (when a 256-vertex block spans >= 2^32 bits)
    uint64_t lo = 0;
    uint64_t base_bits = 0;     // stream bit of device word 0 (device bit positions = stream bits - base_bits)
    uint64_t offs_bytes = 0, word_bytes = 0;  // H2D volume (e2e accounting)
    uint32_t* wbits = nullptr;  // record bits per 32-vertex word (dir_edges), built on the device at load
    Offs offs() const { return Offs{anc, rel, full, lo}; }
};

// Interval checkpoint table of the out-CGR (expand.cuh, Checkpoints), device arrays.
struct DevCk {
    uint32_t *wptr = nullptr, *bits = nullptr, *ck0 = nullptr, *prev = nullptr, *ilen = nullptr;
    uint64_t *after = nullptr, *pos = nullptr;
    IvEntry* q = nullptr;
    uint64_t rows = 0, chunks = 0;
};

struct gcgt_graph {
    int device = 0;
    cudaStream_t stream = nullptr;
    bool own_stream = false;
    cudaStream_t cap_stream = nullptr;  // private stream for graph capture (the caller's may be the legacy stream)
    uint64_t n = 0, nbits = 0, nw = 0;  // nw = words of an n-bit bitmap (padded)
    gcgt_params P{};
    uint64_t lo = 0, hi = 0;
    int rank = 0, nranks = 1;
    DevCgr out, in;
    DevCk ck;
    static constexpr uint32_t kCkC = 3;
    uint32_t ck_c = kCkC;  // intervals per checkpoint chunk (GCGT_TUNE ck_c; 0 = no table).  Vertices with more
                           // intervals hand them to the grid-wide chunk pass (r2 sweep: 32 -> 3 gives C4 20.9 -> 17.7 ms)
    bool in_alias = false;  // symmetric: in == out
    bool has_in = false;
    bool dir_opt = false;
    // uncompressed baseline (gcgt_load_csr, §8 f3)
    bool is_csr = false;
    uint64_t* crow = nullptr;
    uint32_t* ccol = nullptr;
    uint64_t* crow_in = nullptr;
    uint32_t* ccol_in = nullptr;
    bool csr_in_owned = false;
    CsrHubEntry* csr_hubq = nullptr;
    // work buffers
    uint32_t *V = nullptr, *F = nullptr, *N = nullptr;
    uint32_t* q = nullptr;      // BFS: 2 x nw ping-pong word queues; BC: all levels (nw + n)
    uint32_t* qbits = nullptr;  // BC: frontier bits per queue entry
    uint32_t* lvl_off = nullptr;
    LevelState* ls = nullptr;
    HubEntry* hubq = nullptr;
    unsigned long long* hub_ctr = nullptr;   // [0] hub segments, [1] interval chunks (entries << 32 | items)
    unsigned long long* cursor = nullptr;  // [0] work cursor, [1] finished blocks
    unsigned long long* st = nullptr;      // [vertices, arcs, bits]
    unsigned long long* aux = nullptr;     // [4] counters of the partitioned steps (hooks, frontier size, scratch)
    uint32_t* src_dev = nullptr;           // BFS / BC source (graph replay reads it)
    int32_t* levels = nullptr;
    uint32_t* parent = nullptr;
    uint32_t* dirty = nullptr;             // dist CC: changed-parent bitmap
    double *sigma = nullptr, *delta = nullptr, *bc = nullptr, *bcx = nullptr;
    // pinned host mirror (one small block): level state, counters, source
    uint8_t* hp = nullptr;
    LevelState* h_ls() const { return reinterpret_cast<LevelState*>(hp); }
    unsigned long long* h_st() const { return reinterpret_cast<unsigned long long*>(hp + 80); }
    uint32_t* h_src() const { return reinterpret_cast<uint32_t*>(hp + 112); }
    unsigned long long* h_misc() const { return reinterpret_cast<unsigned long long*>(hp + 128); }
    cudaEvent_t ev0 = nullptr, ev1 = nullptr;
    int num_sms = 148;
    // knobs (GCGT_TUNE="key=value,..." at load; results never change)
    uint32_t hub_segs = 1;                  // more segments than this: the vertex's segments go grid-wide
    uint32_t bu_alpha = 30, bu_beta = 128;  // direction switch on vertex counts; alpha in tenths (r2 sweeps, C2-C4)
    uint32_t alpha_bits = 25;               // tenths
    bool bu_grow = false;                   // Beamer's "frontier growing" condition for the switch to bottom-up
                                            // (r2 sweep, alpha 3 without it: C2 4.28, C3 6.55, C4 17.60 ms)
    bool nfilter = false;                   // BFS filter: also test an L1 read of N before the claim
    bool hub_stage = true;                  // hub pass: segments staged through shared memory
    bool dir_bits = false;
    bool dir_edges = true;                  // Beamer's edge rule on CGR bits (DecideArgs::use_edges)
    uint32_t alpha_edges = 0;               // tenths (0: only the guarded second test)
    uint32_t alpha_edges2 = 250;            // tenths; second test, only when nf > edge_guard / 10 * previous nf
    uint32_t edge_guard = 40;               // tenths
    uint64_t in_nbits = 0;                  // bits of the loaded in-records (dir_edges)
    bool dir_opt_knob = true;
    bool use_graph = true;                  // BFS as one CUDA graph (else: chunked host-driven level loop)
    uint32_t chunk = 4;                     // host-driven loop: levels enqueued per host check
    bool compact_offs = true;
    bool td_stage = true;  // top-down: records staged through shared memory with coalesced 128-bit loads
    bool td_pool = true;   // top-down: phase B from a per-warp segment pool, one flat loop with lane refill
                           // (hub_segs capped at 2; r2: C4 BFS 30.1 -> 21.3 ms, C2 7.2 -> 5.7 ms)
    // BFS graph (built on first use for a given levels buffer)
    cudaGraphExec_t bfs_exec = nullptr;
    int32_t* bfs_exec_levels = nullptr;
    // profiling
    bool profile = false, spans = false;
    static constexpr int kKev = 128;
    cudaEvent_t kevp[2 * kKev] = {};
    int kev_n = 0;
    cudaEvent_t sev[5] = {};
    double span_ms[4] = {0, 0, 0, 0};
    double kernel_ms = 0;
    uint64_t kernel_launches = 0;
    uint64_t launches = 0;
    int occ_expand = 0, occ_hub = 0, occ_bu = 0;
};

namespace {

inline int flat_grid(const gcgt_graph* g, uint64_t n) {
    return (int)std::max<uint64_t>(1, std::min<uint64_t>((n + kBlock - 1) / kBlock, (uint64_t)g->num_sms * 16));
}

// The contraction closes each level with one completion atomic per block: 4 blocks per SM keep that serial tail short
// while the dense scan still has 32 warps per SM.
inline int commit_grid(const gcgt_graph* g) {
    return (int)std::max<uint64_t>(1, std::min<uint64_t>((g->nw + kBlock - 1) / kBlock, (uint64_t)g->num_sms * 4));
}

// ---- dispatch over the template parameters (zeta_k, segmented) ------------------------------------------------------
template <class Fn>
inline void with_k(const gcgt_params& P, Fn&& fn) {
    const bool seg = P.residual_segment_len != 0;
#define GCGT_K(KK)                                                      \
    if (seg) fn(std::integral_constant<int, KK>{}, std::true_type{});   \
    else fn(std::integral_constant<int, KK>{}, std::false_type{});
#ifdef GCGT_DEV_K  // development builds (GCGT_DEV_K=3 python -m ...build): one zeta_k only, compiles ~5x faster
    if (P.zeta_k == GCGT_DEV_K) { GCGT_K(GCGT_DEV_K) }
#else
    switch (P.zeta_k) {
        case 1: GCGT_K(1) break;
        case 2: GCGT_K(2) break;
        case 3: GCGT_K(3) break;
        case 4: GCGT_K(4) break;
        default: GCGT_K(5) break;
    }
#endif
#undef GCGT_K
}

template <class T>
inline int occupancy(T kernel) {
    int per_sm = 0;
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kernel, kBlock, 0);
    return std::max(1, per_sm);
}

inline Ctx make_ctx(const gcgt_graph* g) {
    return Ctx{g->out.W, g->out.offs(), g->P.min_interval_len, 8 * g->P.residual_segment_len, g->hub_segs,
               g->hubq, g->hub_ctr, g->st, g->cursor, nullptr, g->td_stage ? kMaxVertexGran : 0u,
               g->td_pool ? 1u : 0u, g->hub_stage ? 1u : 0u,
               Checkpoints{g->ck.wptr, g->ck.bits, g->ck.ck0, g->ck.after, g->ck.pos, g->ck.prev, g->ck.ilen,
                           g->lo >> 5, g->ck_c, g->ck.q, g->hub_ctr + 1}};
}

// Top-down expansion (+ hub pass) of one frontier: a persistent grid at the kernel's occupancy.
template <class App, class Front>
inline void launch_expand(gcgt_graph* g, cudaStream_t s, const Ctx& c, const Front& fr, const App& app,
                          bool reset = true) {
    with_k(g->P, [&](auto KK, auto SS) {
        constexpr int K = decltype(KK)::value;
        constexpr bool SEG = decltype(SS)::value;
        static int occ = 0, occh = 0;
        if (!occ) occ = occupancy(expand_kernel<K, SEG, App, Front>);
        expand_kernel<K, SEG, App, Front><<<occ * g->num_sms, kBlock, 0, s>>>(c, fr, app, 0u);
        g->launches++;
        if (SEG || g->ck.bits) {  // hub segments and / or interval chunks
            if (!occh) occh = occupancy(hub_kernel<K, App>);
            hub_kernel<K, App><<<occh * g->num_sms, kBlock, 0, s>>>(c, app);
            g->launches++;
        }
    });
    if (reset) {  // the work cursor and hub queue for the next launch (the BFS / BC contraction does this itself)
        cudaMemsetAsync(g->cursor, 0, 16, s);
        cudaMemsetAsync(g->hub_ctr, 0, 16, s);
    }
}

inline void launch_bu(gcgt_graph* g, cudaStream_t s, const uint32_t* V, const uint32_t* F, uint32_t* N,
                      uint64_t lo, uint64_t hi, const uint32_t* dir) {
    with_k(g->P, [&](auto KK, auto SS) {
        constexpr int K = decltype(KK)::value;
        constexpr bool SEG = decltype(SS)::value;
        static int occ = 0;
        if (!occ) occ = occupancy(bu_kernel<K, SEG>);
        const uint64_t words = (hi - lo + 31) / 32 + 1;
        const int grid = (int)std::max<uint64_t>(1, std::min<uint64_t>((words + kWarps - 1) / kWarps,
                                                                        (uint64_t)occ * g->num_sms));
        bu_kernel<K, SEG><<<grid, kBlock, 0, s>>>(g->in.W, g->in.offs(), g->P.min_interval_len,
                                                  8 * g->P.residual_segment_len, V, F, N, lo, hi, dir, g->st);
        g->launches++;
    });
}

gcgt_status copy_out(gcgt_graph* g, void* dst, const void* src, size_t bytes, int placement) {
    if (dst == src) return GCGT_OK;
    CU(cudaMemcpyAsync(dst, src, bytes, placement == GCGT_OUT_DEVICE ? cudaMemcpyDeviceToDevice : cudaMemcpyDeviceToHost,
                       g->stream));
    return GCGT_OK;
}

// Brackets one launch of the dominant kernel(s) when profiling: event pairs from a pool, read at the next host sync.
inline gcgt_status kprof_begin(gcgt_graph* g, cudaStream_t s) {
    if (!g->profile) return GCGT_OK;
    if (g->kev_n >= gcgt_graph::kKev) return fail(GCGT_EINVAL, "too many profiled launches between syncs");
    cudaEvent_t& e = g->kevp[2 * g->kev_n];
    if (!e) CU(cudaEventCreate(&e));
    CU(cudaEventRecord(e, s));
    return GCGT_OK;
}
inline gcgt_status kprof_end(gcgt_graph* g, cudaStream_t s) {
    if (!g->profile) return GCGT_OK;
    cudaEvent_t& e = g->kevp[2 * g->kev_n + 1];
    if (!e) CU(cudaEventCreate(&e));
    CU(cudaEventRecord(e, s));
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
    CU(cudaMemsetAsync(g->st, 0, 3 * sizeof(unsigned long long), g->stream));
    CU(cudaEventRecord(g->ev0, g->stream));
    return GCGT_OK;
}

gcgt_status end_call(gcgt_graph* g, gcgt_stats* out, uint32_t iterations) {
    CU(cudaEventRecord(g->ev1, g->stream));
    CU(cudaMemcpyAsync(g->h_st(), g->st, 3 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, g->stream));
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
    if (out) {
        float ms = 0;
        CU(cudaEventElapsedTime(&ms, g->ev0, g->ev1));
        out->iterations = iterations;
        out->reserved = 0;
        out->vertices_expanded = g->h_st()[0];
        out->arcs_decoded = g->h_st()[1];
        out->cgr_bits_decoded = g->h_st()[2];
        out->device_ms = ms;
        out->kernel_ms = g->kernel_ms;
        out->kernel_launches = g->kernel_launches;
        out->launches = g->launches;
    }
    return GCGT_OK;
}

// Small pinned host blocks (per-graph mirrors) are recycled process-wide: cudaFreeHost on every unload measured
// 0.6 ms typical with stalls of 12-314 ms (r1 session 4), inside the bench's end-to-end step.
constexpr size_t kSmallPinned = 256;
std::mutex g_small_mu;
std::vector<void*> g_small_free;
cudaError_t small_pinned_get(void** p) {
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
void small_pinned_put(void* p) {
    if (!p) return;
    std::lock_guard<std::mutex> lk(g_small_mu);
    g_small_free.push_back(p);
}
static_assert(sizeof(LevelState) <= 80, "pinned mirror layout");

// Graph buffers come from the device's stream-ordered memory pool, which keeps freed memory (release threshold =
// max), so repeated load / unload cycles reuse device memory instead of paying cudaMalloc / cudaFree each time.
template <class T>
gcgt_status galloc(const gcgt_graph* g, T** p, uint64_t count) {
    cudaError_t e = cudaMallocAsync((void**)p, std::max<uint64_t>(1, count) * sizeof(T), g->stream);
    if (e != cudaSuccess) return fail(GCGT_ENOMEM, std::string("cudaMallocAsync: ") + cudaGetErrorString(e));
    return GCGT_OK;
}

template <class T>
gcgt_status dalloc(T** p, uint64_t count) {
    cudaError_t e = cudaMalloc((void**)p, std::max<uint64_t>(1, count) * sizeof(T));
    if (e != cudaSuccess) return fail(GCGT_ENOMEM, std::string("cudaMalloc: ") + cudaGetErrorString(e));
    return GCGT_OK;
}

gcgt_cgr_tables* whole_tables(const gcgt_cgr* c) {  // caller holds c->mu
    if (!c->tables) c->tables.reset(new gcgt_cgr_tables());
    return c->tables.get();
}

// Compact bit offsets of vertices [lo, hi): a u64 anchor per 256 vertices (relative to bit `base`) and
// a u32 offset relative to the anchor; t->compact is false when some 256-vertex block spans >= 2^32 bits.
void build_compact(const uint64_t* bo, uint64_t lo, uint64_t hi, uint64_t base, gcgt_cgr_tables* t) {
    const uint64_t nloc = hi - lo, nanc = nloc / 256 + 1;
    bool compact = true;
    for (uint64_t k = 0; compact && k < nanc; k++) {
        const uint64_t a = lo + k * 256, b = std::min(hi, a + 256);
        if (bo[b] - bo[a] >= (1ull << 32)) compact = false;
    }
    t->compact = compact;
    if (!compact) return;
    t->anc.resize(nanc);
    t->rel.resize(nloc + 1);
    uint64_t* anc = t->anc.data();
    uint32_t* rel = t->rel.data();
#pragma omp parallel for schedule(static)
    for (int64_t i = 0; i <= (int64_t)nloc; i++) {
        const uint64_t a = bo[lo + ((uint64_t)i & ~255ull)];
        rel[i] = (uint32_t)(bo[lo + i] - a);
        if ((i & 255) == 0) anc[i >> 8] = a - base;
    }
}

// Uploads the records of vertices [lo, hi) of a host CGR: whole 64-bit stream words (records are self-contained,
// so a vertex-range slice is a bit copy, §8 e) byte-swapped on the device into stream order, plus the bit offsets
// re-based to the slice, in compact form when every 256-vertex block spans < 2^32 bits (§8 a2).  The word array is
// padded so that 128-bit staging loads and the readers' look-ahead never leave it.
gcgt_status upload_cgr(gcgt_graph* g, const gcgt_cgr* c, uint64_t lo, uint64_t hi, bool host_resident, DevCgr* d) {
    cudaStream_t s = g->stream;
    const uint64_t* bo = c->bit_offsets.data() - c->base;  // indexed by global vertex id (slices start at base)
    const uint64_t w0 = bo[lo] / 64;
    const uint64_t wend = (bo[hi] + 63) / 64;
    const uint64_t nwords = ((wend - w0) + 8) & ~1ull;  // >= 6 zero words of padding, even (16-byte granules)
    const uint64_t avail = c->words.size() > w0 ? std::min<uint64_t>(c->words.size() - w0, nwords) : 0;
    gcgt_status st;
    d->lo = lo;
    d->base_bits = w0 * 64;
    d->word_bytes = nwords * 8;
    if (host_resident) {
        CU(cudaHostAlloc((void**)&d->hostW, nwords * sizeof(uint64_t), cudaHostAllocMapped | cudaHostAllocPortable));
        uint64_t* h = d->hostW;
#pragma omp parallel for schedule(static)
        for (int64_t i = 0; i < (int64_t)nwords; i++)
            h[i] = (uint64_t)i < avail ? __builtin_bswap64(c->words[w0 + i]) : 0;
        CU(cudaHostGetDevicePointer((void**)&d->W, h, 0));
    } else {
        if ((st = galloc(g, &d->W, nwords))) return st;
        CU(cudaMemsetAsync(d->W + avail, 0, (nwords - avail) * sizeof(uint64_t), s));
        CU(cudaMemcpyAsync(d->W, c->words.data() + w0, avail * sizeof(uint64_t), cudaMemcpyHostToDevice, s));
        bswap_words<<<flat_grid(g, nwords), kBlock, 0, s>>>(d->W, avail);
    }
    const uint64_t nloc = hi - lo, base = w0 * 64;
    const uint64_t nanc = nloc / 256 + 1;
    const bool whole = lo == c->base && hi == c->base + c->n;  // then base == 0 and the tables are cached
    gcgt_cgr_tables local;
    gcgt_cgr_tables* t = &local;
    std::unique_lock<std::mutex> lk(c->mu, std::defer_lock);
    if (whole) {
        lk.lock();
        t = whole_tables(c);
    }
    if (g->compact_offs && t->anc.empty()) build_compact(bo, lo, hi, base, t);
    if (g->compact_offs && t->compact) {
        if ((st = galloc(g, &d->anc, nanc)) || (st = galloc(g, &d->rel, nloc + 1))) return st;
        CU(cudaMemcpyAsync(d->anc, t->anc.data(), nanc * 8, cudaMemcpyHostToDevice, s));
        CU(cudaMemcpyAsync(d->rel, t->rel.data(), (nloc + 1) * 4, cudaMemcpyHostToDevice, s));
        if (!whole) CU(cudaStreamSynchronize(s));  // local host vectors
        d->offs_bytes = nanc * 8 + (nloc + 1) * 4;
    } else {
        std::vector<uint64_t> ro(nloc + 1);
        for (uint64_t i = 0; i <= nloc; i++) ro[i] = bo[lo + i] - base;
        if ((st = galloc(g, &d->full, nloc + 1))) return st;
        CU(cudaMemcpyAsync(d->full, ro.data(), (nloc + 1) * 8, cudaMemcpyHostToDevice, s));
        CU(cudaStreamSynchronize(s));
        d->offs_bytes = (nloc + 1) * 8;
    }
    const uint64_t nwl = ((hi + 31) >> 5) - (lo >> 5);
    if ((st = galloc(g, &d->wbits, nwl + 1))) return st;
    word_bits_kernel<<<flat_grid(g, nwl), kBlock, 0, s>>>(d->offs(), lo, hi, d->wbits);
    return GCGT_OK;
}

// Upper bound on the vertices whose residual segments go to the hub queue (more than hub_segs segments means a
// record longer than hub_segs * segBits bits): sizes the per-level hub queue without decoding anything.
uint64_t count_hub_bound(const gcgt_cgr* c, uint64_t lo, uint64_t hi, uint64_t min_bits) {
    const uint64_t* bo = c->bit_offsets.data() - c->base;
    uint64_t cnt = 0;
#pragma omp parallel for reduction(+ : cnt) schedule(static)
    for (int64_t u = (int64_t)lo; u < (int64_t)hi; u++) cnt += bo[u + 1] - bo[u] > min_bits;
    return cnt;
}

// Host reader of the canonical MSB-first bytes (FORMAT.md R1), for the load-time checkpoint table only.
struct HostBits {
    const uint8_t* b;
    int bit(uint64_t i) const { return (b[i >> 3] >> (7 - (i & 7))) & 1; }
    uint64_t read(uint32_t K, uint64_t& p) const {  // one VLC codeword (App. B; FORMAT.md R3/R4)
        {  // fast path: a 57+-bit window at p (the words array is padded, so 8 bytes at p/8 are readable)
            uint64_t w;
            memcpy(&w, b + (p >> 3), 8);
            const uint64_t win = __builtin_bswap64(w) << (p & 7);
            if (win) {
                const uint32_t z = (uint32_t)__builtin_clzll(win);
                if (K == 1 && 2 * z + 1 <= 57) {
                    p += 2 * z + 1;
                    return win >> (63 - 2 * z);
                }
                if (K > 1 && (z + 1) * (K + 1) <= 57) {
                    const uint32_t h = z + 1;
                    p += h * (K + 1);
                    return (win << h) >> (64 - K * h);
                }
            }
        }
        uint64_t z = 0;
        while (!bit(p)) { z++; p++; }
        uint64_t payload;
        if (K == 1) payload = z + 1;
        else { p++; payload = (z + 1) * K; }
        uint64_t v = 0;
        for (uint64_t t = 0; t < payload; t++) v = (v << 1) | (uint64_t)bit(p + t);
        p += payload;
        return v;
    }
};

// Interval checkpoint table (expand.cuh, Checkpoints) for the vertices [lo, hi) with more than C intervals: decoded
// on the host (the header of every vertex, the interval area of the few long ones).  Bit positions are relative to
// `base` (the device word array's first bit).
void build_ck_host(const gcgt_cgr* c, uint64_t lo, uint64_t hi, uint64_t base, uint32_t C, gcgt_cgr_tables* t) {
    const uint64_t nloc = hi - lo;
    const uint64_t* bo = c->bit_offsets.data() - c->base;
    const HostBits hb{reinterpret_cast<const uint8_t*>(c->words.data())};
    const bool seg = c->params.residual_segment_len != 0;
    const uint32_t K = c->params.zeta_k;
    t->ck_built = true;
    t->ck_c = C;
    std::vector<uint32_t> itv(nloc, 0);
#pragma omp parallel for schedule(dynamic, 65536)
    for (int64_t i = 0; i < (int64_t)nloc; i++) {
        uint64_t p = bo[lo + i];
        if (p == bo[lo + i + 1]) continue;
        if (!seg) hb.read(K, p);
        const uint64_t x = hb.read(K, p) - 1;
        if (x > C) itv[i] = (uint32_t)x;
    }
    const uint64_t w0 = lo >> 5, nwl = ((hi + 31) >> 5) - w0;
    std::vector<uint32_t> rows_u;
    for (uint64_t i = 0; i < nloc; i++)
        if (itv[i]) rows_u.push_back((uint32_t)(lo + i));
    t->rows = rows_u.size();
    if (rows_u.empty()) return;
    t->wptr.assign(nwl + 1, 0);
    t->bits.assign(nwl, 0);
    for (uint32_t v : rows_u) t->bits[(v >> 5) - w0] |= 1u << (v & 31);
    for (uint64_t w = 0; w < nwl; w++) t->wptr[w + 1] = t->wptr[w] + __builtin_popcount(t->bits[w]);
    const uint64_t R = rows_u.size();
    t->ck0.assign(R + 1, 0);
    t->ilen.assign(R, 0);
    t->after.assign(R, 0);
    for (uint64_t r = 0; r < R; r++) t->ck0[r + 1] = t->ck0[r] + (itv[rows_u[r] - lo] + C - 1) / C;
    const uint64_t T = t->ck0[R];
    t->chunks = T;
    t->pos.assign(T, 0);
    t->prev.assign(T, 0);
#pragma omp parallel for schedule(dynamic, 1)
    for (int64_t r = 0; r < (int64_t)R; r++) {
        const uint64_t u = rows_u[r];
        const uint32_t n_itv = itv[u - lo];
        uint64_t p = bo[u];
        if (!seg) hb.read(K, p);
        hb.read(K, p);
        int64_t prev_end = 0;
        uint64_t sum = 0;
        for (uint32_t k = 0; k < n_itv; k++) {
            if (k % C == 0) {
                t->pos[t->ck0[r] + k / C] = p - base;
                t->prev[t->ck0[r] + k / C] = (uint32_t)prev_end;
            }
            const uint64_t gcode = hb.read(K, p);
            const uint64_t len = hb.read(K, p) - 1 + c->params.min_interval_len;
            int64_t start;
            if (k == 0) {
                const uint64_t z = gcode - 1;
                start = (int64_t)u + ((z & 1) ? -(int64_t)(z >> 1) : (int64_t)(z >> 1));  // R9
            } else {
                start = prev_end + (int64_t)gcode;  // R10
            }
            prev_end = start + (int64_t)len - 1;
            sum += len;
        }
        t->after[r] = p - base;
        t->ilen[r] = (uint32_t)sum;
    }
}

// Uploads the checkpoint table of the owned range (cached with the CGR for whole-CGR loads).
gcgt_status build_checkpoints(gcgt_graph* g, const gcgt_cgr* c) {
    const uint32_t C = g->ck_c;
    if (C == 0 || g->hi == g->lo) return GCGT_OK;
    const bool whole = g->lo == c->base && g->hi == c->base + c->n;
    gcgt_cgr_tables local;
    gcgt_cgr_tables* t = &local;
    std::unique_lock<std::mutex> lk(c->mu, std::defer_lock);
    if (whole) {
        lk.lock();
        t = whole_tables(c);
    }
    if (!t->ck_built || t->ck_c != C) build_ck_host(c, g->lo, g->hi, g->out.base_bits, C, t);
    if (t->rows == 0) return GCGT_OK;
    const uint64_t nwl = t->bits.size(), R = t->rows, T = t->chunks;
    DevCk& d = g->ck;
    gcgt_status st;
    if ((st = galloc(g, &d.wptr, nwl + 1)) || (st = galloc(g, &d.bits, nwl)) || (st = galloc(g, &d.ck0, R + 1)) ||
        (st = galloc(g, &d.after, R)) || (st = galloc(g, &d.ilen, R)) || (st = galloc(g, &d.pos, T)) ||
        (st = galloc(g, &d.prev, T)) || (st = galloc(g, &d.q, R + 1)))
        return st;
    cudaStream_t s = g->stream;
    CU(cudaMemcpyAsync(d.wptr, t->wptr.data(), (nwl + 1) * 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemcpyAsync(d.bits, t->bits.data(), nwl * 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemcpyAsync(d.ck0, t->ck0.data(), (R + 1) * 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemcpyAsync(d.after, t->after.data(), R * 8, cudaMemcpyHostToDevice, s));
    CU(cudaMemcpyAsync(d.ilen, t->ilen.data(), R * 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemcpyAsync(d.pos, t->pos.data(), T * 8, cudaMemcpyHostToDevice, s));
    CU(cudaMemcpyAsync(d.prev, t->prev.data(), T * 4, cudaMemcpyHostToDevice, s));
    if (!whole) CU(cudaStreamSynchronize(s));  // local host vectors
    d.rows = R;
    d.chunks = T;
    return GCGT_OK;
}

void parse_tune(gcgt_graph* g) {
    const char* tune = getenv("GCGT_TUNE");  // development knob: key=value,... (results never change)
    if (!tune) return;
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
            if (k == "hub_segs") g->hub_segs = (uint32_t)std::max(1ul, std::min(8ul, v));
            else if (k == "bu_alpha") g->bu_alpha = (uint32_t)v;
            else if (k == "bu_beta") g->bu_beta = (uint32_t)v;
            else if (k == "dir_bits") g->dir_bits = v != 0;
            else if (k == "alpha_bits") g->alpha_bits = (uint32_t)v;
            else if (k == "dir_edges") g->dir_edges = v != 0;
            else if (k == "alpha_edges") g->alpha_edges = (uint32_t)v;
            else if (k == "alpha_edges2") g->alpha_edges2 = (uint32_t)v;
            else if (k == "edge_guard") g->edge_guard = (uint32_t)v;
            else if (k == "dir_opt") g->dir_opt_knob = v != 0;
            else if (k == "graph") g->use_graph = v != 0;
            else if (k == "chunk") g->chunk = (uint32_t)std::max(2ul, std::min(32ul, v & ~1ul));
            else if (k == "compact") g->compact_offs = v != 0;
            else if (k == "td_stage") g->td_stage = v != 0;
            else if (k == "td_pool") g->td_pool = v != 0;
            else if (k == "ck_c") g->ck_c = (uint32_t)v;
            else if (k == "bu_grow") g->bu_grow = v != 0;
            else if (k == "nfilter") g->nfilter = v != 0;
            else if (k == "hub_stage") g->hub_stage = v != 0;
        }
        i = j + 1;
    }
}

gcgt_status init_graph(gcgt_graph* g, const gcgt_load_opts& o) {
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev == 0) return fail(GCGT_ECUDA, "no CUDA device");
    if (o.device < 0 || o.device >= ndev) return fail(GCGT_EINVAL, "bad device ordinal");
    g->device = o.device;
    CU(cudaSetDevice(o.device));
    {  // keep freed pool memory for the next load (see galloc)
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
    void* hp = nullptr;
    CU(small_pinned_get(&hp));
    g->hp = (uint8_t*)hp;
    CU(cudaEventCreate(&g->ev0));
    CU(cudaEventCreate(&g->ev1));
    for (auto& e : g->sev) CU(cudaEventCreate(&e));
    parse_tune(g);
    if (g->td_pool) g->hub_segs = std::min<uint32_t>(g->hub_segs, 2);  // a pooled round adds <= 32 x 2 tasks
    return GCGT_OK;
}

// Work buffers shared by the CGR and CSR paths.
gcgt_status alloc_work(gcgt_graph* g) {
    gcgt_status st;
    g->nw = ((g->n + 31) / 32 + 1 + 3) & ~3ull;
    if ((st = galloc(g, &g->V, g->nw)) || (st = galloc(g, &g->F, g->nw)) || (st = galloc(g, &g->N, g->nw)) ||
        (st = galloc(g, &g->q, 2 * g->nw)) || (st = galloc(g, &g->ls, 1)) || (st = galloc(g, &g->hub_ctr, 2)) ||
        (st = galloc(g, &g->cursor, 2)) || (st = galloc(g, &g->st, 3)) || (st = galloc(g, &g->src_dev, 1)) ||
        (st = galloc(g, &g->aux, 4)))
        return st;
    CU(cudaMemsetAsync(g->N, 0, g->nw * 4, g->stream));
    CU(cudaMemsetAsync(g->cursor, 0, 16, g->stream));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, g->stream));
    CU(cudaMemsetAsync(g->ls, 0, sizeof(LevelState), g->stream));
    return GCGT_OK;
}

gcgt_status ensure_levels(gcgt_graph* g) {
    if (g->levels) return GCGT_OK;
    return galloc(g, &g->levels, g->n);
}

DecideArgs decide_args(const gcgt_graph* g) {
    return DecideArgs{g->n, g->bu_alpha, g->bu_beta, g->dir_opt ? 1 : 0, g->dir_bits && g->dir_opt ? 1 : 0,
                      (double)g->nbits / (double)std::max<uint64_t>(1, g->n), g->dir_edges ? g->alpha_edges
                                                                                            : g->alpha_bits,
                      g->bu_grow ? 1 : 0, g->dir_edges && g->dir_opt && !g->is_csr ? 1 : 0, (double)g->in_nbits,
                      g->alpha_edges2, g->edge_guard};
}

CommitArgs bfs_commit_args(gcgt_graph* g, int parity, int32_t* lv) {
    CommitArgs a{};
    a.V = g->V;
    a.F = g->F;
    a.N = g->N;
    a.w_lo = 0;
    a.w_hi = g->nw;
    a.qn = g->q + (uint64_t)(1 - parity) * g->nw;
    a.qn_len = &g->ls->qlen[1 - parity];
    a.qcur_len = &g->ls->qlen[parity];
    a.levels = lv;
    a.ls = g->ls;
    a.hub_ctr = g->hub_ctr;
    a.cursor = g->cursor;
    a.dec = decide_args(g);
    a.use_mf = a.dec.use_bits || a.dec.use_edges;
    a.use_mu = a.dec.use_edges;
    if (a.use_mu) {
        a.wb_out = g->out.wbits;
        a.wb_in = g->in.wbits;
    }
    if (a.use_mf && !g->is_csr) a.offs_bits = g->out.offs();
    if (a.use_mf && g->is_csr) a.offs_bits = Offs{nullptr, nullptr, g->crow, 0};
    return a;
}

}  // namespace

// ------------------------------------------------------------------------------------------------------------------
// BFS level enqueue (shared by the host-driven loop and the CUDA-graph body).  Level parity p: the frontier queue is
// q[p] with length ls->qlen[p]; the contraction writes q[1-p].
// ------------------------------------------------------------------------------------------------------------------
namespace {

gcgt_status enqueue_td(gcgt_graph* g, cudaStream_t s, int p) {
    const uint32_t* dir = g->dir_opt ? &g->ls->dir : nullptr;
    const QueueFront fr{g->q + (uint64_t)p * g->nw, &g->ls->qlen[p], g->F, nullptr};
    const BfsApp app{g->V, g->N, g->nfilter ? 1u : 0u};
    if (g->is_csr) {
        static int occ = 0;
        if (!occ) occ = occupancy(csr_expand_kernel<QueueFront>);
        csr_expand_kernel<QueueFront><<<occ * g->num_sms, kBlock, 0, s>>>(g->crow, g->ccol, fr, app, g->cursor,
                                                                          g->csr_hubq, g->hub_ctr, dir, g->st);
        csr_hub_kernel<<<g->num_sms * 4, kBlock, 0, s>>>(g->ccol, g->csr_hubq, g->hub_ctr, app, g->st);
        g->launches += 2;
        return GCGT_OK;
    }
    Ctx c = make_ctx(g);
    c.dir = dir;
    launch_expand(g, s, c, fr, app, false);
    return GCGT_OK;
}

gcgt_status enqueue_bu(gcgt_graph* g, cudaStream_t s) {
    if (g->is_csr) {
        static int occ = 0;
        if (!occ) occ = occupancy(csr_bu_kernel);
        const int grid = (int)std::max<uint64_t>(1, std::min<uint64_t>((g->nw + kWarps - 1) / kWarps,
                                                                        (uint64_t)occ * g->num_sms));
        csr_bu_kernel<<<grid, kBlock, 0, s>>>(g->crow_in, g->ccol_in, g->V, g->F, g->N, g->n, &g->ls->dir, g->st);
        g->launches++;
        return GCGT_OK;
    }
    launch_bu(g, s, g->V, g->F, g->N, 0, g->n, &g->ls->dir);
    return GCGT_OK;
}

gcgt_status enqueue_commit(gcgt_graph* g, cudaStream_t s, int p, int32_t* lv, int use_cond,
                           cudaGraphConditionalHandle cond, int use_dcond, cudaGraphConditionalHandle dcond) {
    CommitArgs a = bfs_commit_args(g, p, lv);
    a.use_cond = use_cond;
    a.cond = cond;
    a.use_dcond = use_dcond;
    a.dcond = dcond;
    commit_kernel<<<commit_grid(g), kBlock, 0, s>>>(a);
    g->launches++;
    return GCGT_OK;
}

// Host-driven level (profiling / tracing / fallback): both directions are launched, each gated on ls->dir.
gcgt_status enqueue_level_host(gcgt_graph* g, int p, int32_t* lv) {
    cudaStream_t s = g->stream;
    gcgt_status st;
    if ((st = kprof_begin(g, s))) return st;
    if (g->spans) CU(cudaEventRecord(g->sev[0], s));
    if ((st = enqueue_td(g, s, p))) return st;
    if (g->spans) CU(cudaEventRecord(g->sev[1], s));
    if (g->spans) CU(cudaEventRecord(g->sev[2], s));
    if (g->dir_opt && (st = enqueue_bu(g, s))) return st;
    if (g->spans) CU(cudaEventRecord(g->sev[3], s));
    if ((st = kprof_end(g, s))) return st;
    return enqueue_commit(g, s, p, lv, 0, 0, 0, 0);
}

// The BFS level loop as one graph: while (frontier non-empty) { level(0); level(1) }, each level an if/else node on
// the direction (bottom-up body | top-down body) followed by the contraction, which sets both conditions.
gcgt_status build_bfs_graph(gcgt_graph* g, int32_t* lv) {
    if (g->bfs_exec) {
        cudaGraphExecDestroy(g->bfs_exec);
        g->bfs_exec = nullptr;
    }
    if (!g->cap_stream) CU(cudaStreamCreateWithFlags(&g->cap_stream, cudaStreamNonBlocking));
    cudaStream_t cs = g->cap_stream;
    cudaGraph_t graph = nullptr;
    CU(cudaGraphCreate(&graph, 0));
    std::unique_ptr<CUgraph_st, cudaError_t (*)(cudaGraph_t)> guard(graph, cudaGraphDestroy);
    cudaGraphConditionalHandle hloop, hdir[2] = {0, 0};
    CU(cudaGraphConditionalHandleCreate(&hloop, graph, 1, cudaGraphCondAssignDefault));
    if (g->dir_opt) {  // (a handle no node uses makes the instantiation fail)
        CU(cudaGraphConditionalHandleCreate(&hdir[0], graph, 0, cudaGraphCondAssignDefault));
        CU(cudaGraphConditionalHandleCreate(&hdir[1], graph, 0, cudaGraphCondAssignDefault));
    }
    cudaGraphNodeParams wp = {};
    wp.type = cudaGraphNodeTypeConditional;
    wp.conditional.handle = hloop;
    wp.conditional.type = cudaGraphCondTypeWhile;
    wp.conditional.size = 1;
    cudaGraphNode_t wnode;
    CU(cudaGraphAddNode(&wnode, graph, nullptr, 0, &wp));
    cudaGraph_t body = wp.conditional.phGraph_out[0];
    cudaGraphNode_t prev = nullptr;
    const uint64_t saved_launches = g->launches;
    for (int p = 0; p < 2; p++) {
        cudaGraphNode_t tail = prev;
        if (g->dir_opt) {  // if/else on the direction the previous contraction chose: [0] bottom-up, [1] top-down
            cudaGraphNodeParams ip = {};
            ip.type = cudaGraphNodeTypeConditional;
            ip.conditional.handle = hdir[p];
            ip.conditional.type = cudaGraphCondTypeIf;
            ip.conditional.size = 2;
            CU(cudaGraphAddNode(&tail, body, prev ? &prev : nullptr, prev ? 1 : 0, &ip));
            cudaGraph_t tmp;
            CU(cudaStreamBeginCaptureToGraph(cs, ip.conditional.phGraph_out[0], nullptr, nullptr, 0,
                                             cudaStreamCaptureModeThreadLocal));
            gcgt_status st = enqueue_bu(g, cs);
            CU(cudaStreamEndCapture(cs, &tmp));
            if (st) return st;
            CU(cudaStreamBeginCaptureToGraph(cs, ip.conditional.phGraph_out[1], nullptr, nullptr, 0,
                                             cudaStreamCaptureModeThreadLocal));
            st = enqueue_td(g, cs, p);
            CU(cudaStreamEndCapture(cs, &tmp));
            if (st) return st;
        }
        // (top-down only: the expansion kernels), then the contraction, which sets the loop / direction conditions
        CU(cudaStreamBeginCaptureToGraph(cs, body, tail ? &tail : nullptr, nullptr, tail ? 1 : 0,
                                         cudaStreamCaptureModeThreadLocal));
        gcgt_status st = g->dir_opt ? GCGT_OK : enqueue_td(g, cs, p);
        if (!st) st = enqueue_commit(g, cs, p, lv, 1, hloop, g->dir_opt ? 1 : 0, hdir[1 - p]);
        // the new tail: the capture's current dependency (the contraction just captured)
        cudaStreamCaptureStatus cst;
        const cudaGraphNode_t* deps = nullptr;
        size_t ndeps = 0;
        const cudaError_t ce = cudaStreamGetCaptureInfo(cs, &cst, nullptr, nullptr, &deps, &ndeps);
        prev = (ce == cudaSuccess && ndeps == 1) ? deps[0] : nullptr;
        cudaGraph_t tmp;
        CU(cudaStreamEndCapture(cs, &tmp));
        if (st) return st;
        CU(ce);
        if (!prev) return fail(GCGT_ECUDA, "graph build: contraction node not found");
    }
    g->launches = saved_launches;
    CU(cudaGraphInstantiate(&g->bfs_exec, graph, 0));
    g->bfs_exec_levels = lv;
    return GCGT_OK;
}

}  // namespace

// ------------------------------------------------------------------------------------------------------------------
// C ABI: load / unload
// ------------------------------------------------------------------------------------------------------------------
extern "C" void gcgt_unload(gcgt_graph* g) {
    if (!g) return;
    cudaSetDevice(g->device);
    if (g->bfs_exec) cudaGraphExecDestroy(g->bfs_exec);
    void* bufs[] = {g->out.hostW ? nullptr : g->out.W, g->out.anc, g->out.rel, g->out.full, g->out.wbits,
                    g->in_alias ? nullptr : g->in.wbits,
                    g->in_alias ? nullptr : (g->in.hostW ? nullptr : g->in.W), g->in_alias ? nullptr : g->in.anc,
                    g->in_alias ? nullptr : g->in.rel, g->in_alias ? nullptr : g->in.full,
                    g->V, g->F, g->N, g->q, g->qbits, g->lvl_off, g->ls, g->hubq, g->hub_ctr, g->cursor, g->st,
                    g->aux, g->ck.wptr, g->ck.bits, g->ck.ck0, g->ck.after,
                    g->ck.ilen, g->ck.pos, g->ck.prev, g->ck.q,
                    g->src_dev, g->levels, g->parent, g->dirty, g->sigma, g->delta, g->bc, g->bcx,
                    g->crow, g->ccol, g->csr_hubq,
                    g->csr_in_owned ? g->crow_in : nullptr, g->csr_in_owned ? g->ccol_in : nullptr};
    if (g->stream) {
        for (void* b : bufs)
            if (b) cudaFreeAsync(b, g->stream);
        cudaStreamSynchronize(g->stream);
    }
    if (g->out.hostW) cudaFreeHost(g->out.hostW);
    if (!g->in_alias && g->in.hostW) cudaFreeHost(g->in.hostW);
    small_pinned_put(g->hp);
    if (g->ev0) cudaEventDestroy(g->ev0);
    if (g->ev1) cudaEventDestroy(g->ev1);
    for (auto& e : g->kevp)
        if (e) cudaEventDestroy(e);
    for (auto& e : g->sev)
        if (e) cudaEventDestroy(e);
    if (g->cap_stream) cudaStreamDestroy(g->cap_stream);
    if (g->own_stream && g->stream) cudaStreamDestroy(g->stream);
    delete g;
}

extern "C" gcgt_status gcgt_load(const gcgt_cgr* c, const gcgt_load_opts* opts, gcgt_graph** out) {
    gcgt_internal::clear_error();
    if (!c || !out) return fail(GCGT_EINVAL, "null argument");
    gcgt_load_opts o{};
    if (opts) o = *opts;
    if (o.nranks > 1 && (o.rank < 0 || o.rank >= o.nranks)) return fail(GCGT_EINVAL, "bad rank");
    if (o.in_cgr) {
        const gcgt_cgr* ic = o.in_cgr;
        if (ic->n_total != c->n_total || ic->base > c->base || ic->base + ic->n < c->base + c->n ||
            ic->params.zeta_k != c->params.zeta_k ||
            ic->params.min_interval_len != c->params.min_interval_len ||
            ic->params.residual_segment_len != c->params.residual_segment_len)
            return fail(GCGT_EINVAL, "in_cgr must have the same n and parameters as the CGR");
    }
    std::unique_ptr<gcgt_graph, void (*)(gcgt_graph*)> g(new gcgt_graph(), gcgt_unload);
    gcgt_status st;
    if ((st = init_graph(g.get(), o))) return st;
    g->n = c->n_total;
    g->nbits = c->nbits;
    g->P = c->params;
    // 1-D vertex-range partition (§8 e): rank r owns [lo, hi), boundaries on 32-vertex words, balanced by CGR bits.
    // A vertex-range slice of a CGR (gcgt_encode_slice) is loaded as exactly its range.
    g->lo = c->base;
    g->hi = c->base + c->n;
    g->nranks = o.nranks > 1 ? o.nranks : 1;
    g->rank = o.nranks > 1 ? o.rank : 0;
    const bool slice = c->base != 0 || c->n != c->n_total;
    if (slice && (c->base % 32 || (g->hi % 32 && g->hi != g->n)))
        return fail(GCGT_EINVAL, "a loaded slice must start and end on 32-vertex words");
    if (slice && g->nranks < 2) g->nranks = 2;  // partitioned: the gcgt_dist_* steps
    if (g->nranks > 1 && !slice) {
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
    }
    if ((st = upload_cgr(g.get(), c, g->lo, g->hi, o.host_resident != 0, &g->out))) return st;
    // in-CGR for bottom-up levels: the transpose's records of the owned vertices, or the CGR itself when symmetric
    if (o.in_cgr) {
        if ((st = upload_cgr(g.get(), o.in_cgr, g->lo, g->hi, o.host_resident != 0, &g->in))) return st;
        g->has_in = true;
        g->in_nbits = o.in_cgr->nbits;
    } else if (o.symmetric) {
        g->in = g->out;
        g->in_alias = true;
        g->has_in = true;
        g->in_nbits = c->nbits;
    }
    g->dir_opt = g->has_in && o.direction_optimizing != 0 && g->dir_opt_knob;
    if ((st = alloc_work(g.get()))) return st;
    const uint64_t seg_bits = 8ull * g->P.residual_segment_len;
    const uint64_t nhub = seg_bits ? count_hub_bound(c, g->lo, g->hi, (uint64_t)g->hub_segs * seg_bits) : 0;
    if ((st = galloc(g.get(), &g->hubq, nhub + 1))) return st;
    if ((st = build_checkpoints(g.get(), c))) return st;
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
    *out = g.release();
    return GCGT_OK;
}

// Uncompressed baseline load (§8 f3): plain CSR on the device; in-lists = the host transpose (counting sort) or the
// CSR itself when symmetric.  Shares the frontier buffers, filter and contraction with the CGR path.
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
    std::unique_ptr<gcgt_graph, void (*)(gcgt_graph*)> g(new gcgt_graph(), gcgt_unload);
    gcgt_status st;
    if ((st = init_graph(g.get(), o))) return st;
    g->is_csr = true;
    g->dir_bits = g->dir_bits || (o.symmetric != 0 && getenv("GCGT_TUNE") == nullptr);
    g->n = n;
    g->lo = 0;
    g->hi = n;
    g->nbits = m;  // the CSR's "record bits" for the direction test: arcs
    cudaStream_t s = g->stream;
    if ((st = galloc(g.get(), &g->crow, n + 1)) || (st = galloc(g.get(), &g->ccol, m))) return st;
    if ((st = alloc_work(g.get()))) return st;
    CU(cudaMemcpyAsync(g->crow, csr->row_offsets, (n + 1) * 8, cudaMemcpyHostToDevice, s));
    if (m) CU(cudaMemcpyAsync(g->ccol, csr->cols, m * 4, cudaMemcpyHostToDevice, s));
    uint64_t nhub = 0;
    for (uint64_t v = 0; v < n; v++) nhub += csr->row_offsets[v + 1] - csr->row_offsets[v] > kCsrHub;
    if ((st = galloc(g.get(), &g->csr_hubq, nhub + 1))) return st;
    if (o.direction_optimizing) {
        if (o.symmetric) {
            g->crow_in = g->crow;
            g->ccol_in = g->ccol;
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
        }
        g->dir_opt = g->dir_opt_knob;
    }
    CU(cudaStreamSynchronize(s));
    CU(cudaGetLastError());
    *out = g.release();
    return GCGT_OK;
}

// ------------------------------------------------------------------------------------------------------------------
// C ABI: queries
// ------------------------------------------------------------------------------------------------------------------
namespace gcgt_internal {
void release_tables(gcgt_cgr* c) {
    std::lock_guard<std::mutex> lk(c->mu);
    if (!c->tables) return;
    for (auto& pr : c->tables->pinned) cudaHostUnregister(pr.first);
    c->tables.reset();
}
}  // namespace gcgt_internal

// Builds the derived load tables of a whole CGR now (compact offsets, checkpoint table for the default chunk size)
// and page-locks the CGR's host arrays, so that every later gcgt_load of it is DMA copies only.
extern "C" gcgt_status gcgt_cgr_pin(gcgt_cgr* c) {
    gcgt_internal::clear_error();
    if (!c) return fail(GCGT_EINVAL, "null argument");
    std::lock_guard<std::mutex> lk(c->mu);
    gcgt_cgr_tables* t = whole_tables(c);
    if (!t->pinned.empty()) return GCGT_OK;
    const uint64_t* bo = c->bit_offsets.data() - c->base;
    if (t->anc.empty()) build_compact(bo, c->base, c->base + c->n, 0, t);
    const uint32_t C = gcgt_graph::kCkC;
    if (!t->ck_built) build_ck_host(c, c->base, c->base + c->n, 0, C, t);
    auto reg = [&](const void* p, size_t bytes) -> gcgt_status {
        if (!p || !bytes) return GCGT_OK;
        const cudaError_t e = cudaHostRegister(const_cast<void*>(p), bytes, cudaHostRegisterPortable);
        if (e != cudaSuccess) return fail(GCGT_ECUDA, std::string("cudaHostRegister: ") + cudaGetErrorString(e));
        t->pinned.emplace_back(const_cast<void*>(p), bytes);
        return GCGT_OK;
    };
    gcgt_status st;
    if ((st = reg(c->words.data(), c->words.size() * 8)) || (st = reg(t->anc.data(), t->anc.size() * 8)) ||
        (st = reg(t->rel.data(), t->rel.size() * 4)) || (st = reg(t->pos.data(), t->pos.size() * 8)) ||
        (st = reg(t->prev.data(), t->prev.size() * 4)))
        return st;
    if (!t->compact && (st = reg(c->bit_offsets.data(), c->bit_offsets.size() * 8))) return st;
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

extern "C" gcgt_status gcgt_bfs(gcgt_graph* g, uint32_t source, int32_t* levels, int placement, gcgt_stats* stats) {
    if (!g || !levels) return fail(GCGT_EINVAL, "null argument");
    if (g->nranks > 1) return fail(GCGT_EINVAL, "partitioned graph: use the gcgt_dist_* steps (dist.py)");
    if (source >= g->n) return fail(GCGT_ERANGE, "source >= n");
    gcgt_status st;
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    int32_t* lv = levels;
    if (placement != GCGT_OUT_DEVICE) {
        if ((st = ensure_levels(g))) return st;
        lv = g->levels;
    }
    *g->h_src() = source;
    CU(cudaMemcpyAsync(g->src_dev, g->h_src(), 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->F, 0, g->nw * 4, s));
    seed_kernel<<<1, 1, 0, s>>>(g->src_dev, g->V, g->F, g->q, nullptr, lv, g->ls, nullptr, nullptr);
    g->launches = 1;
    const bool graph = g->use_graph && !g->profile;
    if (graph) {
        if (!g->bfs_exec || g->bfs_exec_levels != lv) {
            if ((st = build_bfs_graph(g, lv))) return st;
        }
        CU(cudaGraphLaunch(g->bfs_exec, s));
        g->launches++;
        CU(cudaMemcpyAsync(g->h_ls(), g->ls, sizeof(LevelState), cudaMemcpyDeviceToHost, s));
    } else {
        // Host-driven level loop without a per-level wait: kernels size their work from the device-resident state, so
        // the host enqueues `chunk` levels (an even number: the queue parity restarts at 0) and checks for an empty
        // frontier once per chunk; levels enqueued past the end find an empty queue and exit at once.  Span
        // profiling (gcgt_profile(g, 2)) waits per level.
        for (uint32_t level = 0;;) {
            const uint32_t nlev = g->spans ? 2 : std::min<uint32_t>(g->chunk, gcgt_graph::kKev);
            for (uint32_t i = 0; i < nlev; i++, level++) {
                if ((st = enqueue_level_host(g, (int)(level & 1), lv))) return st;
                if (g->spans) {
                    CU(cudaEventRecord(g->sev[4], s));
                    CU(cudaEventSynchronize(g->sev[4]));
                    float lms[4];
                    for (int k = 0; k < 4; k++) {
                        CU(cudaEventElapsedTime(&lms[k], g->sev[k], g->sev[k + 1]));
                        g->span_ms[k] += lms[k];
                    }
                    if (getenv("GCGT_TRACE")) {  // development aid (tools/trace_bfs.py): one line per level
                        LevelState h;
                        CU(cudaMemcpy(&h, g->ls, sizeof(h), cudaMemcpyDeviceToHost));
                        fprintf(stderr, "level %3u next_dir %u visited %10u new %9u next_words %8u | exp %.4f "
                                "bu %.4f commit %.4f ms\n", level, h.dir, h.visited, h.prev_nf, h.qlen[(level + 1) & 1],
                                lms[0], lms[2], lms[3]);
                    }
                }
            }
            CU(cudaMemcpyAsync(g->h_ls(), g->ls, sizeof(LevelState), cudaMemcpyDeviceToHost, s));
            CU(cudaStreamSynchronize(s));
            if ((st = kprof_collect(g))) return st;
            if (g->h_ls()->qlen[level & 1] == 0) break;
        }
    }
    finalize_levels<<<flat_grid(g, (g->n + 31) / 32), kBlock, 0, s>>>(g->V, lv, g->n);
    g->launches++;
    if ((st = copy_out(g, levels, lv, g->n * 4, placement))) return st;
    if ((st = end_call(g, stats, 0))) return st;
    if (stats) {
        const LevelState* h = g->h_ls();
        stats->iterations = h->nonempty + 1;  // non-empty levels (the seed level included)
        if (graph) {  // kernels the graph ran: per level the expansion kernel(s) of its direction + the contraction
            const uint32_t td_kernels = g->is_csr ? 2 : ((g->P.residual_segment_len || g->ck.bits) ? 2 : 1);
            stats->launches += (uint64_t)h->ntd * td_kernels + h->nbu + h->ntd + h->nbu;
        }
    }
    return GCGT_OK;
}

// Weakly connected components: one hooking pass of the expansion engine over every vertex (CcApp), then pointer
// jumping (the CAS hooking never overwrites a link, so one pass suffices).
extern "C" gcgt_status gcgt_cc(gcgt_graph* g, uint32_t* labels, int placement, gcgt_stats* stats) {
    if (!g || !labels) return fail(GCGT_EINVAL, "null argument");
    if (g->is_csr) return fail(GCGT_EINVAL, "CSR baseline graph: BFS only");
    if (g->nranks > 1) return fail(GCGT_EINVAL, "partitioned graph: use the gcgt_dist_* steps (dist.py)");
    gcgt_status st;
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    uint32_t* lab = placement == GCGT_OUT_DEVICE ? labels : nullptr;
    if (!lab) {
        if (!g->parent && (st = galloc(g, &g->parent, g->n))) return st;
        lab = g->parent;
    }
    cc_init<<<flat_grid(g, g->n), kBlock, 0, s>>>(lab, g->n);
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    const Ctx c = make_ctx(g);
    const DenseFront fr{g->lo, g->hi};
    const CcApp app{lab, nullptr, nullptr, 0, 0};  // single GPU: no hook counting
    if ((st = kprof_begin(g, s))) return st;
    launch_expand(g, s, c, fr, app);
    if ((st = kprof_end(g, s))) return st;
    cc_jump<<<flat_grid(g, g->n), kBlock, 0, s>>>(lab, g->n);
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    g->launches += 2;
    if ((st = copy_out(g, labels, lab, g->n * 4, placement))) return st;
    CU(cudaStreamSynchronize(s));
    if ((st = kprof_collect(g))) return st;
    return end_call(g, stats, 1);
}

// Betweenness centrality (Brandes): per source a forward pass (sigma) whose levels are kept in one all-levels queue,
// then the backward pass (delta) over the levels in reverse.  The forward loop runs without per-level host round
// trips (the level state is on the device); the host reads the level offsets once per source.
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
            (st = galloc(g, &g->bcx, g->n)) ||
            (st = galloc(g, &g->qbits, g->n + g->nw)) || (st = galloc(g, &g->lvl_off, g->n + 3 + 2 * gcgt_graph::kKev)))
            return st;
        uint32_t* bigq = nullptr;
        if ((st = galloc(g, &bigq, g->n + g->nw))) return st;
        cudaFreeAsync(g->q, g->stream);
        g->q = bigq;
        g->bfs_exec_levels = nullptr;  // the BFS graph captured the old queue pointer
        if (g->bfs_exec) {
            cudaGraphExecDestroy(g->bfs_exec);
            g->bfs_exec = nullptr;
        }
    }
    if ((st = ensure_levels(g))) return st;
    if ((st = begin_call(g))) return st;
    cudaStream_t s = g->stream;
    const Ctx c = make_ctx(g);
    CU(cudaMemsetAsync(g->bc, 0, g->n * 8, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    std::vector<uint32_t> lvl_off;
    for (uint32_t si = 0; si < k; si++) {
        *g->h_src() = sources[si];
        CU(cudaMemcpyAsync(g->src_dev, g->h_src(), 4, cudaMemcpyHostToDevice, s));
        CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
        CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
        CU(cudaMemsetAsync(g->sigma, 0, g->n * 8, s));
        CU(cudaMemsetAsync(g->delta, 0, g->n * 8, s));
        seed_kernel<<<1, 1, 0, s>>>(g->src_dev, g->V, nullptr, g->q, g->qbits, g->levels, g->ls, g->lvl_off, g->sigma);
        // forward: the level's queue range is read from the device state (ls->q_off, q_len)
        for (uint32_t level = 0;;) {
            for (uint32_t i = 0; i < g->chunk; i++, level++) {
                const QueueFront fr{g->q, &g->ls->q_len, nullptr, g->qbits, &g->ls->q_off};
                const BcFwdApp app{g->V, g->N, g->sigma, 0.0};
                if ((st = kprof_begin(g, s))) return st;
                launch_expand(g, s, c, fr, app, false);
                if ((st = kprof_end(g, s))) return st;
                CommitArgs a{};
                a.V = g->V;
                a.N = g->N;
                a.w_lo = 0;
                a.w_hi = g->nw;
                a.qn = g->q;
                a.qbits = g->qbits;
                a.lvl_off = g->lvl_off;
                a.levels = g->levels;
                a.ls = g->ls;
                a.hub_ctr = g->hub_ctr;
                a.cursor = g->cursor;
                a.bc = 1;
                commit_kernel<<<commit_grid(g), kBlock, 0, s>>>(a);
                g->launches++;
            }
            CU(cudaMemcpyAsync(g->h_ls(), g->ls, sizeof(LevelState), cudaMemcpyDeviceToHost, s));
            CU(cudaStreamSynchronize(s));
            if ((st = kprof_collect(g))) return st;
            if (g->h_ls()->q_len == 0) break;
        }
        const uint32_t D = g->h_ls()->nonempty + 1;  // levels 0..D-1
        lvl_off.resize(D + 1);
        CU(cudaMemcpyAsync(lvl_off.data(), g->lvl_off, (D + 1) * 4, cudaMemcpyDeviceToHost, s));
        CU(cudaStreamSynchronize(s));
        for (int d = (int)D - 2; d >= 0; d--) {  // the last level has no successors
            const uint32_t off = lvl_off[d];
            const uint32_t off1 = lvl_off[d + 1], len1 = lvl_off[d + 2] - off1;  // level d+1's queue range
            bc_level_bits<<<flat_grid(g, len1), kBlock, 0, s>>>(g->q + off1, g->qbits + off1, len1, g->N, 1);
            bc_level_x<<<flat_grid(g, (uint64_t)len1 * 32), kBlock, 0, s>>>(g->q + off1, g->qbits + off1, len1,
                                                                            g->sigma, g->delta, g->bcx);
            const QueueFront fr{g->q + off, nullptr, nullptr, g->qbits + off, nullptr, lvl_off[d + 1] - off};
            const BcBwdApp app{g->N, g->bcx, g->sigma, g->delta, g->bc, sources[si], 0, 0.0};
            launch_expand(g, s, c, fr, app);
            CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
            bc_level_bits<<<flat_grid(g, len1), kBlock, 0, s>>>(g->q + off1, g->qbits + off1, len1, g->N, 0);
            g->launches += 3;
        }
    }
    if ((st = copy_out(g, bc, g->bc, g->n * 8, placement))) return st;
    return end_call(g, stats, k);
}

// ------------------------------------------------------------------------------------------------------------------
// Partitioned (multi-GPU) steps.  The caller (paper_conf_sigmod_shalt19_b200/dist.py) runs the collectives between
// them; all bitmaps crossing the boundary are device arrays of ceil(n/32) 32-bit words (bit v%32 of word v/32).
// Every step is enqueued on the graph's stream and returns without waiting, except those that hand a count to the
// host (gcgt_dist_bfs_absorb, gcgt_dist_cc_hook): one host sync per BFS level / CC round.
// ------------------------------------------------------------------------------------------------------------------
extern "C" gcgt_status gcgt_dist_bfs_begin(gcgt_graph* g, uint32_t source) {
    gcgt_internal::clear_error();
    if (!g) return fail(GCGT_EINVAL, "null graph");
    if (g->is_csr) return fail(GCGT_EINVAL, "CSR baseline graph: single-GPU BFS only");
    if (source >= g->n) return fail(GCGT_ERANGE, "source >= n");
    gcgt_status st;
    CU(cudaSetDevice(g->device));
    if ((st = ensure_levels(g))) return st;
    cudaStream_t s = g->stream;
    *g->h_src() = source;
    CU(cudaMemcpyAsync(g->src_dev, g->h_src(), 4, cudaMemcpyHostToDevice, s));
    CU(cudaMemsetAsync(g->V, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->F, 0, g->nw * 4, s));
    CU(cudaMemsetAsync(g->levels, 0xff, g->n * 4, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    seed_kernel<<<1, 1, 0, s>>>(g->src_dev, g->V, g->F, g->q, nullptr, g->levels, g->ls, nullptr, nullptr);
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_bfs_expand(gcgt_graph* g, uint32_t level, uint32_t* cand, uint32_t* fslice,
                                            int bottom_up) {
    gcgt_internal::clear_error();
    if (!g || (bottom_up ? !fslice : !cand)) return fail(GCGT_EINVAL, "null argument");
    if (bottom_up && !g->has_in) return fail(GCGT_EINVAL, "bottom-up needs an in-CGR (or a symmetric graph)");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    (void)level;
    const uint64_t nwf = (g->n + 31) / 32;
    if (bottom_up) {
        // the owned unvisited vertices scan their in-records against the replicated frontier F; finds go straight to
        // the owned slice of the next frontier (no exchange needed before the all-gather)
        const uint64_t w_lo = g->lo / 32, nlw = (g->hi + 31) / 32 - w_lo;
        CU(cudaMemsetAsync(fslice, 0, nlw * 4, s));
        static uint32_t* one = nullptr;  // a device "1": the bottom-up kernel's direction gate
        if (!one) {
            CU(cudaMalloc(&one, 4));
            const uint32_t v = 1;
            CU(cudaMemcpy(one, &v, 4, cudaMemcpyHostToDevice));
        }
        launch_bu(g, s, g->V, g->F, fslice - w_lo, g->lo, g->hi, one);
        return GCGT_OK;
    }
    CU(cudaMemsetAsync(cand, 0, nwf * 4, s));
    const Ctx c = make_ctx(g);
    const BitsFront fr{g->F, g->lo, g->hi};
    const BfsApp app{g->V, cand, g->nfilter ? 1u : 0u};
    launch_expand(g, s, c, fr, app);
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_bfs_commit(gcgt_graph* g, uint32_t level, const uint32_t* recv, uint32_t nparts,
                                            uint32_t* fslice, int keep) {
    gcgt_internal::clear_error();
    if (!g || !fslice || (nparts && !recv)) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    const uint64_t w_lo = g->lo / 32, nlw = (g->hi + 31) / 32 - w_lo;
    unsigned long long* cnt = g->aux + 2;  // scratch counter (new owned vertices; not returned)
    *reinterpret_cast<int32_t*>(g->h_misc()) = (int32_t)level;
    CU(cudaMemcpyAsync(g->src_dev, g->h_misc(), 4, cudaMemcpyHostToDevice, s));
    if (nlw)
        dist_commit<<<flat_grid(g, nlw * 32), kBlock, 0, s>>>(recv, nparts, w_lo, nlw, g->V, fslice, g->levels,
                                                               reinterpret_cast<const int32_t*>(g->src_dev), g->n,
                                                               cnt, keep);
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_bfs_absorb(gcgt_graph* g, const uint32_t* frontier, uint64_t* count) {
    gcgt_internal::clear_error();
    if (!g || !frontier || !count) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    const uint64_t nwf = (g->n + 31) / 32;
    unsigned long long* cnt = g->aux + 1;
    CU(cudaMemsetAsync(cnt, 0, 8, s));
    dist_absorb<<<flat_grid(g, nwf), kBlock, 0, s>>>(frontier, g->F, g->V, nwf, cnt);
    CU(cudaMemcpyAsync(g->h_st() + 1, cnt, 8, cudaMemcpyDeviceToHost, s));
    CU(cudaStreamSynchronize(s));
    CU(cudaGetLastError());
    *count = g->h_st()[1];
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_bfs_levels(gcgt_graph* g, int32_t* levels_owned, int placement) {
    gcgt_internal::clear_error();
    if (!g || !levels_owned) return fail(GCGT_EINVAL, "null argument");
    gcgt_status st;
    if ((st = copy_out(g, levels_owned, g->levels + g->lo, (g->hi - g->lo) * 4, placement))) return st;
    CU(cudaStreamSynchronize(g->stream));
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_cc_hook(gcgt_graph* g, uint32_t* parent, uint32_t* pairs, uint64_t cap,
                                         uint64_t* hooks) {
    gcgt_internal::clear_error();
    if (!g || !parent || !hooks || (cap && !pairs)) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cudaStream_t s = g->stream;
    uint32_t* hc = reinterpret_cast<uint32_t*>(g->aux);  // not the stats block: the engine adds its counts there
    CU(cudaMemsetAsync(hc, 0, 4, s));
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    const Ctx c = make_ctx(g);
    const DenseFront fr{g->lo, g->hi};
    const CcDistApp app{parent, hc, pairs, (uint32_t)std::min<uint64_t>(cap, 0xFFFFFFFFull), 0};
    launch_expand(g, s, c, fr, app);
    CU(cudaMemsetAsync(g->hub_ctr, 0, 16, s));
    CU(cudaMemcpyAsync(g->h_misc(), hc, 4, cudaMemcpyDeviceToHost, s));
    CU(cudaStreamSynchronize(s));
    CU(cudaGetLastError());
    *hooks = *reinterpret_cast<uint32_t*>(g->h_misc());
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_cc_merge(gcgt_graph* g, uint32_t* parent, const uint32_t* pairs, uint64_t npairs) {
    gcgt_internal::clear_error();
    if (!g || !parent || (npairs && !pairs)) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    if (npairs) cc_merge_pairs<<<flat_grid(g, npairs), kBlock, 0, g->stream>>>(parent, pairs, npairs);
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_dist_cc_jump(gcgt_graph* g, uint32_t* parent) {
    gcgt_internal::clear_error();
    if (!g || !parent) return fail(GCGT_EINVAL, "null argument");
    CU(cudaSetDevice(g->device));
    cc_jump<<<flat_grid(g, g->n), kBlock, 0, g->stream>>>(parent, g->n);
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_sync(gcgt_graph* g) {
    gcgt_internal::clear_error();
    if (!g) return fail(GCGT_EINVAL, "null graph");
    CU(cudaStreamSynchronize(g->stream));
    CU(cudaGetLastError());
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

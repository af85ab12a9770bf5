// expand.cuh — top-down frontier expansion over the CGR (expansion + filtering of §6), B200 form.
//
// Work distribution.  A persistent grid (one wave at the occupancy limit) whose warps take batches of frontier
// queue words from an atomic cursor (the first batch of every warp is static, so small frontiers pay no cursor
// atomics).  Within a batch the frontier vertices are listed and processed 32 at a time ("rounds"):
//
//  1. Staging.  Each lane's vertex record [bit_offsets[u], bit_offsets[u+1]) is rounded to 16-byte granules and the
//     warp copies all 32 records into its shared-memory buffer with coalesced 128-bit loads (stage_ranges), so the
//     record misses of the round overlap instead of forming one dependent chain per lane (the uncoalesced,
//     divergent bit-array reads of lane-per-node decoding that §5.1, names as the weakness).
//  2. Phase A (lane per vertex): the record header and the interval area (Alg. 2 l.1-32, :650-688), decoded from
//     shared memory; each interval is claimed as a word range (the Two-Phase "expand a long run in parallel" idea at
//     word granularity: 32 ids per operation).  Then segNum (Fig. 6, :1057-1069).
//  3. Phase B: the round's residual segments — self-contained by R17 ("breaks the sequential dependencies",
//     :945-946) — become tasks of a per-warp pool (default, `pool`): once it holds >= kPoolFlush tasks it is drained by
//     ONE flat loop with lane refill (drain_pool), four neighbour ids per step and lane, so no lane waits for the
//     longest segment of a round.  (pool = 0: the round's segments one per lane from shared memory.)  A vertex with
//     more than hub_segs segments (default 1) hands them to the level's hub queue instead, and a vertex with more than
//     ck_c intervals (default 3) its interval chunks to the chunk queue; the hub pass spreads both over the whole grid
//     (Task Stealing + Residual Segmentation, §4.3/§5.2, at grid scale).
#pragma once
#include "apps.cuh"

namespace gcgt_dev {

struct HubEntry {
    uint64_t base;  // bit position of the vertex's first residual segment
    uint64_t end;   // end of the vertex record
    uint32_t u;
    uint32_t seg_off;  // first flattened segment index (entries are ordered by seg_off)
    uint32_t nseg;
    uint32_t pad;
};

// Long interval areas.  A record with more than ck_c intervals decodes them as one serial chain (each gap is relative to
// the previous interval's end, R10), which on a social hub (10^5 intervals) is milliseconds of one lane.  The load
// step therefore builds a checkpoint table (the residual-segment idea of §5.2, :1092-1136, applied to intervals as a
// derived device table; the CGR bytes are unchanged): for every such vertex, the bit position and the previous
// interval end of every ck_c-th interval, and the position after the interval area.  The expansion hands the
// vertex's interval chunks to the level's chunk queue, which the hub pass spreads over the grid like segments.
struct IvEntry {
    uint32_t u, ck0, nck, off;  // vertex, first checkpoint, chunks, first flattened chunk index
    uint32_t itv, pad;
};

struct Checkpoints {
    const uint32_t* __restrict__ wptr;  // per owned 32-vertex word: table rows before it
    const uint32_t* __restrict__ bits;  // per owned word: which of its vertices have a row
    const uint32_t* __restrict__ ck0;   // per row: first checkpoint (rows + 1 entries)
    const uint64_t* __restrict__ after; // per row: bit position after the interval area
    const uint64_t* __restrict__ pos;   // per checkpoint: bit position of the chunk's first gap code
    const uint32_t* __restrict__ prev;  // per checkpoint: end of the interval before the chunk
    const uint32_t* __restrict__ ilen;  // per row: total interval length (unsegmented records: residual count)
    uint64_t w0;                        // first owned word
    uint32_t ck_c;                      // intervals per chunk; rows exist for vertices with more than ck_c
    IvEntry* q;                         // per-level chunk queue
    unsigned long long* ctr;            // (entries << 32) | chunks
};

// Kernel-constant view of the device CGR plus the per-level hub queue.
struct Ctx {
    const uint64_t* __restrict__ W;
    Offs offs;
    uint32_t min_len, seg_bits, hub_segs;
    HubEntry* hubq;
    unsigned long long* hub_ctr;  // (entries << 32) | segments
    unsigned long long* st;       // [vertices, arcs, bits] counters
    unsigned long long* cursor;   // [0] work cursor over the frontier queue, [1] finished-warp count
    const uint32_t* dir;          // BFS direction gate: top-down kernels run only while *dir == 0 (nullptr: always)
    uint32_t max_gran;            // records staged through shared memory up to this many granules (0: none)
    uint32_t pool;                // phase B from a per-warp task pool filled over several rounds (lane refill)
    uint32_t hub_stage;           // hub pass: segments staged through shared memory
    Checkpoints ck;               // long interval areas (ck.bits == nullptr: none)
};

// ---- frontier sources ------------------------------------------------------------------------------------------------
// Queue of frontier words (BFS / BC): entry i is word q[off + i]; its bits come from qbits[off + i] (BC keeps them
// per level) or from the frontier bitmap F (BFS; the contraction rewrites F densely every level).  The length is
// read from device memory (qlen_p, written by the previous contraction) or given (len); the offset likewise (off_p:
// BC's all-levels queue, advanced on the device).
struct QueueFront {
    const uint32_t* __restrict__ q;
    const uint32_t* __restrict__ qlen_p;
    const uint32_t* __restrict__ F;
    const uint32_t* __restrict__ qbits;
    const uint32_t* __restrict__ off_p;
    uint32_t len;
    __device__ __forceinline__ uint64_t size() const { return qlen_p ? *(volatile const uint32_t*)qlen_p : len; }
    __device__ __forceinline__ void get(uint64_t i, uint32_t& w, uint32_t& bits) const {
        if (off_p) i += *off_p;
        w = q[i];
        bits = qbits ? qbits[i] : F[w];
    }
};

// Frontier bits of the owned word range (partitioned BFS): entry i is word lo/32 + i, restricted to [lo, hi).
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

// One residual segment (FORMAT.md R17): count, the first residual anchored at u, then gaps.  Ids go to the filter
// four at a time so that their probes are in flight together.  Returns the count.
template <int K, class R, class T>
__device__ __forceinline__ uint32_t decode_segment(R& r, uint32_t u, T& t) {
    const uint32_t cnt = (uint32_t)(r.template next<K>() - 1);
    uint32_t cur = 0, done = 0;
    for (; done + 4 <= cnt; done += 4) {  // whole batches of four: no per-id predicates
        uint32_t v[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            const uint64_t c = r.template next<K>();
            cur = (done + k == 0) ? unmap_first32(u, c) : cur + (uint32_t)c;
            v[k] = cur;
        }
        t.many(v, 4);
    }
    if (done < cnt) {  // tail of 1..3
        uint32_t v[4];
        const uint32_t nb = cnt - done;
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            if (k < nb) {
                const uint64_t c = r.template next<K>();
                cur = (done + k == 0) ? unmap_first32(u, c) : cur + (uint32_t)c;
            }
            v[k] = cur;
        }
        t.many(v, nb);
    }
    return cnt;
}

constexpr int kStageGran = 128;  // staging granules (16 B) per warp: 2 KB
constexpr uint32_t kMaxVertexGran = 64;  // records above 8 Kbit are read from global memory
constexpr uint32_t kPool = 160;   // phase-B task pool (segments of several rounds) per warp
constexpr uint32_t kPoolFlush = kPool - 32 * 2;  // a round adds at most 32 x hub_segs (<= 2 when pooling) tasks

struct ExpSmem {
    uint4 stage[kStageGran];
    StageSlots sl;
    uint8_t owner[256];
    uint32_t w[32], b[32], pre[33];
    uint32_t su[32], spre[33];
    uint64_t sbase[32];
    uint64_t tpos[kPool];
    uint32_t tu[kPool];
    uint32_t ntask, take;
};

// Phase B from the pool: every lane takes the next segment task as soon as it finishes one (lane refill from a
// shared-memory cursor), so a round's long segment no longer idles the other lanes; segments are read from global
// memory (the pool outlives the round's staged records).
// The drain is ONE flat loop (no per-segment inner loop, whose reconvergence would make every lane wait for the
// longest segment): each iteration every busy lane decodes up to four residuals of its segment and hands them to the
// filter; lanes whose segment ended take the next pool task (warp-synchronous assignment in pool order).
template <int K, class App>
__device__ __forceinline__ void drain_pool(const Ctx& c, const App& app, ExpSmem& sm, uint32_t& na) {
    const uint32_t lane = lane_id();
    const uint32_t N = sm.ntask;
    const uint32_t* W32 = reinterpret_cast<const uint32_t*>(c.W);
    GBitReader r;
    uint32_t u = 0, rem = 0, cur = 0;
    bool first = false;
    uint32_t next = 0;
    for (;;) {
        const uint32_t need = __ballot_sync(0xffffffffu, rem == 0);
        if (rem == 0) {
            const uint32_t k = next + __popc(need & lanemask_lt());
            if (k < N) {
                u = sm.tu[k];
                r.init(W32, 0, sm.tpos[k]);
                rem = (uint32_t)(r.template next<K>() - 1);
                first = true;
            }
        }
        next += __popc(need);
        if (!__any_sync(0xffffffffu, rem != 0)) break;
        const uint32_t nb = min(rem, 4u);
        uint32_t v[4];
#pragma unroll
        for (uint32_t k = 0; k < 4; k++) {
            if (k < nb) {
                const uint64_t cd = r.template next<K>();
                cur = (k == 0 && first) ? unmap_first32(u, cd) : cur + (uint32_t)cd;
            }
            v[k] = cur;
        }
        first = false;
        App t = app;
        t.begin(u);
        t.many(v, nb);
        t.end();
        rem -= nb;
        na += nb;
    }
    __syncwarp();
    if (lane == 0) sm.ntask = 0;
    __syncwarp();
}

__device__ __forceinline__ void lane_source(const ExpSmem& sm, const uint64_t* W, uint32_t o, const uint32_t*& src,
                                            uint64_t& j0) {
    const uint32_t ex = sm.sl.excl[o];
    if (ex != 0xFFFFFFFFu) {
        src = reinterpret_cast<const uint32_t*>(sm.stage) + (size_t)ex * 4;
        j0 = sm.sl.g0[o] * 4;
    } else {
        src = reinterpret_cast<const uint32_t*>(W);
        j0 = 0;
    }
}

template <int K, bool SEG, class App, class Front>
__device__ __forceinline__ void expand_body(const Ctx& c, const Front& fr, const App& app, uint32_t wpb, ExpSmem& sm,
                                            uint32_t& nv, uint32_t& na, uint32_t& nb) {
    const uint32_t wid = threadIdx.x >> 5, lane = lane_id();
    const uint64_t qlen = fr.size();
    if (wpb == 0) {  // sized on the device (host did not wait for the queue length): ~4 batches per resident warp
        const uint64_t b = qlen / ((uint64_t)gridDim.x * kWarps * 4);
        wpb = b < 1 ? 1 : (b > 8 ? 8 : (uint32_t)b);
    }
    const uint64_t nstatic = (uint64_t)gridDim.x * kWarps * wpb;
    unsigned long long next = ((uint64_t)blockIdx.x * kWarps + wid) * wpb;
    if (SEG && c.pool) {
        if (lane == 0) sm.ntask = 0;
        __syncwarp();
    }
    for (;;) {
        const uint64_t base = __shfl_sync(0xffffffffu, next, 0);
        if (base >= qlen) break;
        if (lane == 0) next = nstatic + atomicAdd(c.cursor, (unsigned long long)wpb);
        uint32_t w = 0, bits = 0;
        if (lane < wpb && base + lane < qlen) fr.get(base + lane, w, bits);
        const uint32_t incl = warp_incl_scan(__popc(bits));
        sm.w[lane] = w;
        sm.b[lane] = bits;
        sm.pre[lane + 1] = incl;
        if (lane == 0) sm.pre[0] = 0;
        __syncwarp();
        const uint32_t total = sm.pre[32];
        for (uint32_t t0 = 0; t0 < total; t0 += 32) {
            const uint32_t j = t0 + lane;
            const bool active = j < total;
            uint32_t u = 0;
            uint64_t p0 = 0, p1 = 0;
            if (active) {
                uint32_t lo = 0, hi = 31;  // owner word: largest o with pre[o] <= j
                while (lo < hi) {
                    const uint32_t mid = (lo + hi + 1) >> 1;
                    if (sm.pre[mid] <= j) lo = mid; else hi = mid - 1;
                }
                u = sm.w[lo] * 32 + __fns(sm.b[lo], 0, (int)(j - sm.pre[lo]) + 1);
                p0 = c.offs(u);
                p1 = c.offs(u + 1);
            }
            sm.sl.excl[lane] = 0xFFFFFFFFu;
            const uint32_t* src;
            uint64_t j0;
            stage_ranges<kStageGran>(reinterpret_cast<uint32_t*>(sm.stage), sm.owner, sm.sl, c.W, active, p0, p1,
                                     c.max_gran, src, j0);
            uint32_t nseg = 0;
            uint64_t sbase = 0;
            if (active) {
                App t = app;
                t.begin(u);
                t.vertex(u);
                nv++;
                nb += (uint32_t)(p1 - p0);
                BitReader r;
                r.init(src, j0, p0);
                uint64_t deg = 0;
                if (!SEG) deg = r.template next<K>() - 1;
                uint32_t itv = (uint32_t)(r.template next<K>() - 1);
                uint32_t prev_end = 0, in_itv = 0;
                if (itv > c.ck.ck_c && c.ck.bits) {  // long interval area: its chunks go grid-wide
                    const uint64_t wl = (u >> 5) - c.ck.w0;
                    const uint32_t row = c.ck.wptr[wl] + __popc(c.ck.bits[wl] & ((1u << (u & 31)) - 1));
                    const uint32_t k0 = c.ck.ck0[row], nck = c.ck.ck0[row + 1] - k0;
                    const unsigned long long old = atomicAdd(c.ck.ctr, (1ull << 32) | (unsigned long long)nck);
                    c.ck.q[old >> 32] = IvEntry{u, k0, nck, (uint32_t)(old & 0xffffffffu), itv, 0};
                    r.init(r.src, r.j0, c.ck.after[row]);
                    itv = 0;
                    in_itv = c.ck.ilen[row];  // counted as arcs by the chunk pass, not here
                    na -= in_itv;
                }
                for (uint32_t i = 0; i < itv; i++) {
                    const uint64_t g = r.template next<K>();
                    const uint32_t len = (uint32_t)(r.template next<K>() - 1) + c.min_len;
                    const uint32_t start = i == 0 ? unmap_first32(u, g) : prev_end + (uint32_t)g;
                    t.range(start, len);
                    prev_end = start + len - 1;
                    in_itv += len;
                }
                na += in_itv;
                if (!SEG) {  // unsegmented record (R8): the residual list, lane-serially
                    const uint32_t nres = (uint32_t)(deg - in_itv);
                    uint32_t cur = 0;
                    for (uint32_t done = 0; done < nres; done += 4) {
                        uint32_t v[4];
                        const uint32_t k_n = min(4u, nres - done);
#pragma unroll
                        for (uint32_t k = 0; k < 4; k++) {
                            if (k < k_n) {
                                const uint64_t cd = r.template next<K>();
                                cur = (done + k == 0) ? unmap_first32(u, cd) : cur + (uint32_t)cd;
                            }
                            v[k] = cur;
                        }
                        t.many(v, k_n);
                    }
                    na += nres;
                } else {
                    nseg = (uint32_t)(r.template next<K>() - 1);
                    sbase = r.pos();
                    if (nseg > c.hub_segs) {  // hub: hand the segments to the whole grid
                        const unsigned long long old = atomicAdd(c.hub_ctr, (1ull << 32) | (unsigned long long)nseg);
                        c.hubq[old >> 32] = HubEntry{sbase, p1, u, (uint32_t)(old & 0xffffffffu), nseg, 0};
                        nseg = 0;
                    }
                }
                t.end();
            }
            if (SEG && c.pool) {
                // ---- phase B (pooled): queue the round's segments; drain when the pool is nearly full
                const uint32_t sincl = warp_incl_scan(nseg);
                const uint32_t n0 = sm.ntask;
                for (uint32_t k = 0; k < nseg; k++) {
                    sm.tu[n0 + sincl - nseg + k] = u;
                    sm.tpos[n0 + sincl - nseg + k] = sbase + (uint64_t)k * c.seg_bits;
                }
                __syncwarp();
                if (lane == 31) sm.ntask = n0 + sincl;
                __syncwarp();
                if (sm.ntask >= kPoolFlush) drain_pool<K>(c, app, sm, na);
            } else if (SEG) {
                // ---- phase B: the round's residual segments, one per lane
                const uint32_t sincl = warp_incl_scan(nseg);
                sm.su[lane] = u;
                sm.sbase[lane] = sbase;
                sm.spre[lane + 1] = sincl;
                if (lane == 0) sm.spre[0] = 0;
                for (uint32_t k = sincl - nseg; k < sincl; k++) sm.owner[k] = (uint8_t)lane;
                __syncwarp();
                const uint32_t S = sm.spre[32];
                for (uint32_t k = lane; k < S; k += 32) {
                    const uint32_t o = sm.owner[k];
                    const uint32_t su = sm.su[o];
                    const uint32_t* s2;
                    uint64_t j2;
                    lane_source(sm, c.W, o, s2, j2);
                    BitReader r;
                    r.init(s2, j2, sm.sbase[o] + (uint64_t)(k - sm.spre[o]) * c.seg_bits);
                    App t = app;
                    t.begin(su);
                    na += decode_segment<K>(r, su, t);
                    t.end();
                }
            }
            __syncwarp();
        }
        __syncwarp();
    }
    if (SEG && c.pool && sm.ntask) drain_pool<K>(c, app, sm, na);
}

template <int K, bool SEG, class App, class Front>
__global__ void __launch_bounds__(kBlock, 5) expand_kernel(Ctx c, Front fr, App app, uint32_t wpb) {
    __shared__ ExpSmem smem[kWarps];
    uint32_t nv = 0, na = 0, nb = 0;
    if (!(c.dir && *c.dir)) expand_body<K, SEG, App, Front>(c, fr, app, wpb, smem[threadIdx.x >> 5], nv, na, nb);
    add_stats3(c.st, nv, na, nb);
    // the work cursor is reset by the next contraction (or a memset by the caller): no per-block completion atomic
}

// ---- hub pass: the level's hub segments flattened over the whole grid -----------------------------------------------
// A warp takes 32 consecutive flattened segments (usually 32 neighbouring segments of one hub, i.e. one contiguous
// 1 KB run of fixed-stride segments, R16), finds their entries with one 32-ary ballot search, stages them with
// coalesced 128-bit loads and decodes one segment per lane from shared memory.
__device__ __forceinline__ uint32_t entry_off(const HubEntry& e) { return e.seg_off; }
__device__ __forceinline__ uint32_t entry_off(const IvEntry& e) { return e.off; }

template <class E>
__device__ __forceinline__ uint32_t warp_find_entry(const E* __restrict__ q, uint32_t ne, uint32_t jb, uint32_t j) {
    const uint32_t lane = lane_id();
    uint32_t lo = 0, hi = ne;  // invariant: off[lo] <= jb, and off[hi] > jb if hi < ne
    while (hi - lo > 1) {
        const uint32_t span = hi - lo;
        const uint32_t pos = span <= 32 ? lo + lane : lo + (uint32_t)(((uint64_t)span * lane) >> 5);
        const bool le = (span > 32 || lane < span) && entry_off(q[pos]) <= jb;
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
    while (e + 1 < ne && entry_off(q[e + 1]) <= j) e++;
    return e;
}

__device__ __forceinline__ uint32_t warp_find_hub(const HubEntry* __restrict__ q, uint32_t ne, uint32_t jb,
                                                  uint32_t j) {
    return warp_find_entry(q, ne, jb, j);
}

// The level's interval chunks (long interval areas, see Checkpoints): one chunk of ck_c intervals per lane, decoded from
// its checkpoint and claimed as word ranges.
template <int K, class App>
__device__ __forceinline__ void chunk_pass(const Ctx& c, const App& app, uint32_t& na) {
    const unsigned long long cc = *(volatile unsigned long long*)c.ck.ctr;
    if (!cc) return;
    const uint32_t lane = lane_id();
    const uint32_t ne = (uint32_t)(cc >> 32), S = (uint32_t)(cc & 0xffffffffu);
    const uint64_t gw0 = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) & ~31ull;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t jb = gw0; jb < S; jb += stride) {
        const uint32_t j = (uint32_t)jb + lane;
        const uint32_t k = warp_find_entry(c.ck.q, ne, (uint32_t)jb, min(j, S - 1));
        if (j >= S) continue;
        const IvEntry e = c.ck.q[k];
        const uint32_t idx = j - e.off, ck = e.ck0 + idx;
        const uint32_t cnt = min(c.ck.ck_c, e.itv - idx * c.ck.ck_c);
        GBitReader r;
        r.init(reinterpret_cast<const uint32_t*>(c.W), 0, c.ck.pos[ck]);
        uint32_t prev_end = c.ck.prev[ck];
        App t = app;
        t.begin(e.u);
        for (uint32_t i = 0; i < cnt; i++) {
            const uint64_t g = r.template next<K>();
            const uint32_t len = (uint32_t)(r.template next<K>() - 1) + c.min_len;
            const uint32_t start = (idx == 0 && i == 0) ? unmap_first32(e.u, g) : prev_end + (uint32_t)g;
            t.range(start, len);
            prev_end = start + len - 1;
            na += len;
        }
        t.end();
    }
}

constexpr int kHubGran = 192;

struct HubSmem {
    uint4 stage[kHubGran];
    StageSlots sl;
    uint8_t owner[kHubGran];
};

template <int K, class App>
__global__ void __launch_bounds__(kBlock) hub_kernel(Ctx c, App app) {
    __shared__ HubSmem smem[kWarps];
    if (c.dir && *c.dir) return;  // a bottom-up level (host-driven loop)
    uint32_t na = 0;
    if (c.ck.bits) chunk_pass<K>(c, app, na);
    const unsigned long long hc = *(volatile unsigned long long*)c.hub_ctr;
    if (hc == 0) {  // no hub segments this level
        add_stats3(c.st, 0, na, 0);
        return;
    }
    HubSmem& sm = smem[threadIdx.x >> 5];
    const uint32_t lane = lane_id();
    const uint32_t nh = (uint32_t)(hc >> 32), S = (uint32_t)(hc & 0xffffffffu);
    const uint64_t gw0 = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) & ~31ull;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t jb = gw0; jb < S; jb += stride) {
        const uint32_t j = (uint32_t)jb + lane;
        const bool active = j < S;
        const uint32_t k = warp_find_hub(c.hubq, nh, (uint32_t)jb, min(j, S - 1));
        uint64_t q = 0, qe = 0;
        uint32_t u = 0;
        if (active) {
            const HubEntry e = c.hubq[k];
            const uint32_t sidx = j - e.seg_off;
            u = e.u;
            q = e.base + (uint64_t)sidx * c.seg_bits;
            qe = sidx + 1 == e.nseg ? e.end : q + c.seg_bits;
        }
        const uint32_t* src;
        uint64_t j0;
        stage_ranges<kHubGran>(reinterpret_cast<uint32_t*>(sm.stage), sm.owner, sm.sl, c.W, active, q, qe,
                               c.hub_stage ? 32u : 0u, src, j0);
        if (active) {
            BitReader r;
            r.init(src, j0, q);
            App t = app;
            t.begin(u);
            na += decode_segment<K>(r, u, t);
            t.end();
        }
        __syncwarp();
    }
    add_stats3(c.st, 0, na, 0);
}

}  // namespace gcgt_dev

// decode.cuh — device-side CGR decoding for sm_100a (FORMAT.md R1-R19).
//
// The device keeps the CGR as 64-bit words in stream order (bit i of the stream is bit 63-(i%64) of word i/64;
// the load step byte-swaps the canonical MSB-first bytes once).  A codeword at bit p is decoded from a 64-bit
// window W[p/64] << (p%64) | W[p/64+1] >> (64 - p%64): one CLZ gives the unary part (App. B),
// one shift pair gives the payload.  gamma codes longer than 63 bits and zeta codes longer than 64 bits take a
// (never-taken on our workloads) slow path.
#pragma once
#include <stdint.h>

namespace gcgt_dev {

__device__ __forceinline__ uint64_t ldg64(const uint64_t* p) { return __ldg(reinterpret_cast<const unsigned long long*>(p)); }

__device__ __forceinline__ uint64_t window(const uint64_t* __restrict__ W, uint64_t p) {
    const uint64_t i = p >> 6;
    const uint32_t s = (uint32_t)(p & 63);
    const uint64_t a = ldg64(W + i), b = ldg64(W + i + 1);
    return s ? (a << s) | (b >> (64 - s)) : a;
}

__device__ __forceinline__ int stream_bit(const uint64_t* __restrict__ W, uint64_t p) {
    return (int)((ldg64(W + (p >> 6)) >> (63 - (p & 63))) & 1);
}

// Slow path: codes whose length exceeds the 64-bit window (gamma >= 64 bits: x >= 2^32; zeta: x >= 2^48).
template <int K>
__device__ __noinline__ uint64_t decode_slow(const uint64_t* __restrict__ W, uint64_t& p) {
    uint64_t z = 0;
    while (!stream_bit(W, p)) { z++; p++; }
    uint64_t payload;
    if (K == 1) payload = z + 1;
    else { p++; payload = (z + 1) * K; }
    uint64_t x = 0;
    for (uint64_t i = 0; i < payload; i++) x = (x << 1) | (uint64_t)stream_bit(W, p + i);
    p += payload;
    return x;
}

// decodeNum (Alg. 1 l.6): one VLC codeword at p; advances p.
// Fast path in 32-bit arithmetic: the top 32 bits of the window (one funnel shift of the two words holding it) hold
// every codeword of at most 32 bits (zeta_3: values < 2^24; gamma: < 2^15), i.e. nearly all gaps and counts; longer
// codewords take the 64-bit window, then the bit-serial slow path.
template <int K>
__device__ __forceinline__ uint64_t decode(const uint64_t* __restrict__ W, uint64_t& p) {
    const uint64_t i = p >> 6;
    const uint32_t s = (uint32_t)(p & 63);
    const uint64_t a = ldg64(W + i), b = ldg64(W + i + 1);
    const uint32_t x = s < 32 ? (uint32_t)(a >> 32) : (uint32_t)a;
    const uint32_t y = s < 32 ? (uint32_t)a : (uint32_t)(b >> 32);
    const uint32_t hi = __funnelshift_l(y, x, s & 31);  // window bits 0..31
    const uint32_t z = __clz(hi);
    if (K == 1) {
        if (z < 16) {
            const uint32_t L = 2 * z + 1;
            p += L;
            return hi >> (32 - L);
        }
    } else {
        const uint32_t h = z + 1, L = h * (K + 1);
        if (L <= 32) {
            p += L;
            return (hi << h) >> (32 - K * h);
        }
    }
    const uint64_t win = s ? (a << s) | (b >> (64 - s)) : a;
    const uint32_t zz = (uint32_t)__clzll((long long)win);
    if (K == 1) {
        if (zz < 32) {
            const uint32_t L = 2 * zz + 1;
            p += L;
            return win >> (64 - L);
        }
    } else {
        const uint32_t h = zz + 1, L = h * (K + 1);
        if (L <= 64) {
            p += L;
            return (win << h) >> (64 - K * h);
        }
    }
    return decode_slow<K>(W, p);
}

// Inverse of the first-gap sign map + 1 (App. C :2101-2106, FORMAT.md R9/R11/R17): code c -> u + delta.
__device__ __forceinline__ int64_t unmap_first(uint64_t u, uint64_t c) {
    const uint64_t z = c - 1;
    return (int64_t)u + ((z & 1) ? -(int64_t)(z >> 1) : (int64_t)(z >> 1));
}

// Walks u's record: calls vis.range(start, len) per interval and vis.one(v) per residual.
// Unsegmented (SEG=false): R8-R12.  Segmented (SEG=true): R14-R17.  Returns the neighbour count.
template <int K, bool SEG, class Visitor>
__device__ __forceinline__ uint32_t walk_record(const uint64_t* __restrict__ W, uint64_t p, uint64_t u,
                                                uint32_t min_len, uint32_t seg_bits, Visitor& vis) {
    uint64_t deg = 0;
    if (!SEG) deg = decode<K>(W, p) - 1;
    const uint64_t itv = decode<K>(W, p) - 1;
    uint64_t got = 0;
    int64_t prev_end = 0;
    for (uint64_t t = 0; t < itv; t++) {
        const uint64_t g = decode<K>(W, p);
        const uint64_t len = decode<K>(W, p) - 1 + min_len;
        const int64_t start = t == 0 ? unmap_first(u, g) : prev_end + (int64_t)g;
        vis.range((uint32_t)start, (uint32_t)len);
        prev_end = start + (int64_t)len - 1;
        got += len;
    }
    if (!SEG) {
        const uint64_t nres = deg - got;
        int64_t cur = 0;
        for (uint64_t t = 0; t < nres; t++) {
            const uint64_t c = decode<K>(W, p);
            cur = t == 0 ? unmap_first(u, c) : cur + (int64_t)c;
            vis.one((uint32_t)cur);
        }
        return (uint32_t)deg;
    } else {
        const uint64_t nseg = decode<K>(W, p) - 1;
        const uint64_t base = p;
        for (uint64_t s = 0; s < nseg; s++) {
            uint64_t q = base + s * seg_bits;
            const uint64_t cnt = decode<K>(W, q) - 1;
            int64_t cur = unmap_first(u, decode<K>(W, q));
            vis.one((uint32_t)cur);
            for (uint64_t t = 1; t < cnt; t++) {
                cur += (int64_t)decode<K>(W, q);
                vis.one((uint32_t)cur);
            }
            got += cnt;
        }
        return (uint32_t)got;
    }
}

}  // namespace gcgt_dev

namespace gcgt_dev {

// Speculative decode for the warp-parallel decoder: the codeword's length, or 0xFFFF when it does not fit the
// 64-bit window path (then only the exact slow path can decode it).
template <int K>
__device__ __forceinline__ uint32_t spec_decode(const uint64_t* __restrict__ W, uint64_t q, uint64_t& val) {
    const uint64_t win = window(W, q);
    const uint32_t z = (uint32_t)__clzll((long long)win);
    if (K == 1) {
        if (z < 32) {
            const uint32_t L = 2 * z + 1;
            val = win >> (64 - L);
            return L;
        }
    } else {
        const uint32_t h = z + 1, L = h * (K + 1);
        if (L <= 64) {
            val = (win << h) >> (64 - K * h);
            return L;
        }
    }
    val = 0;
    return 0xFFFFu;
}

// One window step of Alg. 4 parallelDecode, B200 form, over WIN <= 32 lanes: lane i decodes
// speculatively at p+i (lines 5-7); the valid starts are marked from lane 0 by pointer jumping (lines 9-15,
// Fig. 5): each marked lane marks the start its pointer names (__reduce_or_sync of one-hot masks), then every
// pointer jumps to its target's pointer; 'x' (>= WIN) propagates.  By Lemma 5.2 five rounds cover 32 lanes.
// Returns the mask of lanes holding a valid codeword start; val/len are the lane's speculative decode.
// With TRACE, trace_pos/trace_flags receive the per-round state (row 0 = initial) and *rounds the row count.
template <int K, int WIN, bool TRACE>
__device__ __forceinline__ uint32_t window_step(const uint64_t* __restrict__ W, uint64_t p, uint64_t& val,
                                                uint32_t& len, uint32_t* trace_pos = nullptr,
                                                uint32_t* trace_flags = nullptr, uint32_t* rounds = nullptr) {
    const uint32_t lane = threadIdx.x & 31;
    len = spec_decode<K>(W, p + lane, val);
    uint32_t pos = lane < (uint32_t)WIN ? lane + len : 0xFFFFFFFFu;  // start of the following codeword
    uint32_t flags = 1u;                                             // lane 0 starts a codeword (line 8)
    if (TRACE && lane < (uint32_t)WIN) { trace_pos[lane] = pos; trace_flags[lane] = lane == 0; }
    int r = 0;
#pragma unroll
    for (; r < 5; r++) {
        const uint32_t mark = (((flags >> lane) & 1u) && pos < (uint32_t)WIN) ? (1u << pos) : 0u;
        const uint32_t m = __reduce_or_sync(0xffffffffu, mark);
        if (!m) break;  // line 12: no marked lane points inside the window
        flags |= m;
        const uint32_t pp = __shfl_sync(0xffffffffu, pos, pos & 31);
        pos = pos < (uint32_t)WIN ? pp : 0xFFFFFFFFu;
        if (TRACE && lane < (uint32_t)WIN) {
            trace_pos[(r + 1) * 32 + lane] = pos;
            trace_flags[(r + 1) * 32 + lane] = (flags >> lane) & 1u;
        }
    }
    if (TRACE && lane == 0) *rounds = (uint32_t)r + 1;
    return flags;
}

// Decodes `count` consecutive codewords from bit p with the whole warp (window_step per 32 bits).  The first
// min(#valid, remaining) codewords of each step are handed to fn(step_base, take, index, value, active)
// warp-uniformly (lines 16-17).  Returns the bit after the last codeword.  All 32 lanes must call it with
// warp-uniform p and count.
template <int K, class Fn>
__device__ __forceinline__ uint64_t warp_decode(const uint64_t* __restrict__ W, uint64_t p, uint64_t count, Fn&& fn) {
    const uint32_t lane = threadIdx.x & 31;
    uint32_t lt;
    asm("mov.u32 %0, %%lanemask_lt;" : "=r"(lt));
    uint64_t done = 0;
    while (done < count) {
        uint64_t val;
        uint32_t len;
        const uint32_t flags = window_step<K, 32, false>(W, p, val, len);
        const uint64_t rem = count - done;
        const uint32_t nvalid = __popc(flags);
        const uint32_t take = (uint64_t)nvalid < rem ? nvalid : (uint32_t)rem;
        const uint32_t last = (uint32_t)__fns(flags, 0, (int)take);
        uint32_t last_len = __shfl_sync(0xffffffffu, len, last);
        if (last_len == 0xFFFFu) {  // only the last valid codeword can be this long: decode it exactly
            uint64_t q = p + last;
            const uint64_t v = decode_slow<K>(W, q);
            if (lane == last) val = v;
            last_len = (uint32_t)(q - (p + last));
        }
        const uint32_t idx = __popc(flags & lt);
        const bool act = ((flags >> lane) & 1u) && idx < take;
        fn(done, take, done + idx, val, act);
        p += last + last_len;
        done += take;
    }
    return p;
}

}  // namespace gcgt_dev

namespace gcgt_dev {

// Register-staged bit reader: a 256-bit window (four 64-bit stream words) held in registers and refilled with
// four independent loads when a codeword may cross its end.  Decoding is then pure ALU work (CLZ + shifts):
// one memory round trip per ~256 bits instead of one (L1) round trip per codeword.  Codewords longer than the
// 64-bit path use the global-memory slow path.
struct RegStream {
    const uint64_t* __restrict__ W;
    uint64_t p;      // absolute bit position of the next codeword
    uint64_t base;   // word index of r0
    uint64_t r0, r1, r2, r3;

    __device__ __forceinline__ void fill(uint64_t wi) {
        base = wi;
        r0 = ldg64(W + wi);
        r1 = ldg64(W + wi + 1);
        r2 = ldg64(W + wi + 2);
        r3 = ldg64(W + wi + 3);
    }
    __device__ __forceinline__ void init(const uint64_t* __restrict__ w, uint64_t pos) {
        W = w;
        p = pos;
        fill(pos >> 6);
    }
    __device__ __forceinline__ void seek(uint64_t pos) {
        p = pos;
        const uint64_t wi = pos >> 6;
        if (wi < base || wi + 1 > base + 3) fill(wi);
    }
    __device__ __forceinline__ uint64_t win() {
        uint64_t wi = p >> 6;
        if (wi + 1 > base + 3) {  // the 64-bit window would leave the staged words
            fill(wi);
        }
        const uint32_t k = (uint32_t)(wi - base), s = (uint32_t)(p & 63);
        const uint64_t a = k == 0 ? r0 : k == 1 ? r1 : r2;
        const uint64_t b = k == 0 ? r1 : k == 1 ? r2 : r3;
        return s ? (a << s) | (b >> (64 - s)) : a;
    }
    template <int K>
    __device__ __forceinline__ uint64_t next() {
        const uint64_t w = win();
        const uint32_t z = (uint32_t)__clzll((long long)w);
        if (K == 1) {
            if (z < 32) {
                const uint32_t L = 2 * z + 1;
                p += L;
                return w >> (64 - L);
            }
        } else {
            const uint32_t h = z + 1, L = h * (K + 1);
            if (L <= 64) {
                p += L;
                return (w << h) >> (64 - K * h);
            }
        }
        const uint64_t v = decode_slow<K>(W, p);
        return v;
    }
};

}  // namespace gcgt_dev

namespace gcgt_dev {

// Sequential bit-buffer reader: the next stream bits left-aligned in a 64-bit register, refilled 32 bits at a
// time (32-bit stream word j is ((const uint32_t*)W)[j ^ 1] because W holds 64-bit words in stream order on a
// little-endian machine).  Per codeword: CLZ, two shifts, a length check and an occasional 32-bit load, all in
// 32-bit-friendly arithmetic.  Codewords longer than the buffered bits take the global slow path.
struct BitBuf {
    uint64_t buf;    // next bits, MSB first
    uint32_t avail;  // valid bits in buf
    uint64_t nxt;    // next 32-bit stream word to load

    __device__ __forceinline__ static uint32_t ld32(const uint64_t* __restrict__ W, uint64_t j) {
        return __ldg(reinterpret_cast<const unsigned int*>(W) + (j ^ 1));
    }
    __device__ __forceinline__ void init(const uint64_t* __restrict__ W, uint64_t p) {
        const uint64_t j = p >> 5;
        const uint32_t off = (uint32_t)(p & 31);
        buf = (((uint64_t)ld32(W, j) << 32) | ld32(W, j + 1)) << off;
        avail = 64 - off;
        nxt = j + 2;
    }
    __device__ __forceinline__ uint64_t pos() const { return nxt * 32 - avail; }
    template <int K>
    __device__ __forceinline__ uint64_t next(const uint64_t* __restrict__ W) {
        if (avail <= 32) {
            buf |= (uint64_t)ld32(W, nxt) << (32 - avail);
            avail += 32;
            nxt++;
        }
        // fast path (32-bit arithmetic): after the refill avail > 32, so a codeword of <= 32 bits is complete
        const uint32_t hi = (uint32_t)(buf >> 32);
        const uint32_t z32 = __clz(hi);
        if (K == 1) {
            if (z32 < 16) {
                const uint32_t L = 2 * z32 + 1;
                buf <<= L;
                avail -= L;
                return hi >> (32 - L);
            }
        } else {
            const uint32_t h = z32 + 1, L = h * (K + 1);
            if (L <= 32) {
                buf <<= L;
                avail -= L;
                return (hi << h) >> (32 - K * h);
            }
        }
        const uint32_t z = (uint32_t)__clzll((long long)buf);
        uint32_t L, h = 0;
        if (K == 1) L = 2 * z + 1;
        else { h = z + 1; L = h * (K + 1); }
        if (L < 64 && L <= avail) {
            const uint64_t v = K == 1 ? buf >> (64 - L) : (buf << h) >> (64 - K * h);
            buf <<= L;
            avail -= L;
            return v;
        }
        uint64_t p = pos();  // long codeword (e.g. a segment's first residual): 64-bit window path, then re-seat
        const uint64_t v = decode<K>(W, p);
        init(W, p);
        return v;
    }
};

}  // namespace gcgt_dev

// device.cuh — shared device building blocks of the sm_100a path: lane helpers, fire-and-forget reductions, the
// compact bit-offset table, the CGR bit reader, and the warp-cooperative record staging into shared memory.
//
// CGR words on the device: the canonical MSB-first byte stream (FORMAT.md R1) byte-swapped once at load into 64-bit
// stream words (bit i of the stream = bit 63 - i%64 of word i/64).  As 32-bit words in memory the stream word j is
// ((const uint32_t*)W)[j ^ 1] (little-endian halves), so a 16-byte granule copied verbatim keeps that layout.
#pragma once
#include <stdint.h>

#include "decode.cuh"

namespace gcgt_dev {

constexpr int kBlock = 256;
constexpr int kWarps = kBlock / 32;

__device__ __forceinline__ uint32_t lane_id() { return threadIdx.x & 31; }
__device__ __forceinline__ uint32_t lanemask_lt() {
    uint32_t m;
    asm("mov.u32 %0, %%lanemask_lt;" : "=r"(m));
    return m;
}

// Fire-and-forget reductions (REDG): the claim's old value is never needed, so no round trip to L2 is waited for.
__device__ __forceinline__ void red_or(uint32_t* p, uint32_t v) {
    asm volatile("red.relaxed.gpu.global.or.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ void red_add(unsigned long long* p, unsigned long long v) {
    asm volatile("red.relaxed.gpu.global.add.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void red_add(uint32_t* p, uint32_t v) {
    asm volatile("red.relaxed.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

__device__ __forceinline__ uint32_t warp_incl_scan(uint32_t x) {
    const uint32_t lane = lane_id();
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        const uint32_t t = __shfl_up_sync(0xffffffffu, x, o);
        if (lane >= (uint32_t)o) x += t;
    }
    return x;
}

// Bit offsets of the (owned) vertex records, FORMAT.md R2 (`bitStart[u]`, Alg. 1 l.5).  Compact
// form: a u64 anchor per 256 vertices plus a u32 offset relative to it, 4.03 B per vertex instead of
// 8 (used when every 256-vertex block spans < 2^32 bits); otherwise the plain u64 table.  Indices are relative to
// the owned range's first vertex lo.
struct Offs {
    const uint64_t* __restrict__ anc;
    const uint32_t* __restrict__ rel;
    const uint64_t* __restrict__ full;
    uint64_t lo;
    __device__ __forceinline__ uint64_t operator()(uint64_t v) const {
        const uint64_t i = v - lo;
        if (full) return ldg64(full + i);
        return ldg64(anc + (i >> 8)) + (uint64_t)__ldg(rel + i);
    }
};

// Codeword at bit p of a 32-bit word stream (element 0 = stream word j0): the general path for codewords longer than
// 32 bits (a segment's first residual anchored at u, App. C) and, bit-serially, longer than 64 bits.  Out of line:
// the reader's fast path stays small.
struct Decoded {
    uint64_t v;
    uint64_t end;
};
template <int K, bool GENERIC>
__device__ __forceinline__ Decoded decode_at(const uint32_t* src, uint64_t j0, uint64_t p) {
    auto ld = [&](uint64_t i) { return GENERIC ? src[i ^ 1] : __ldg(src + (i ^ 1)); };
    const uint64_t i = (p >> 5) - j0;
    const uint32_t s = (uint32_t)(p & 31);
    const uint64_t a = ((uint64_t)ld(i) << 32) | ld(i + 1), b = ld(i + 2);
    const uint64_t win = s ? (a << s) | (b << s >> 32) : a;
    const uint32_t z = (uint32_t)__clzll((long long)win);
    if (K == 1 && z < 32) {
        const uint32_t L = 2 * z + 1;
        return Decoded{win >> (64 - L), p + L};
    }
    if (K > 1 && (z + 1) * (K + 1) <= 64) {
        const uint32_t h = z + 1;
        return Decoded{(win << h) >> (64 - K * h), p + h * (K + 1)};
    }
    auto bit = [&](uint64_t q) { return (ld((q >> 5) - j0) >> (31 - (q & 31))) & 1u; };
    uint64_t q = p, zz = 0;
    while (!bit(q)) { zz++; q++; }
    uint64_t payload;
    if (K == 1) payload = zz + 1;
    else { q++; payload = (zz + 1) * K; }
    uint64_t v = 0;
    for (uint64_t t = 0; t < payload; t++) v = (v << 1) | bit(q + t);
    return Decoded{v, q + payload};
}

// Sequential CGR reader over 32-bit stream words: the next stream bits MSB-aligned in two 32-bit registers (hi, lo),
// refilled 32 bits at a time.  Every shift is a 32-bit funnel shift (SHF, one instruction; the 64-bit variable
// shifts they replace cost ~5 each).  Invariant: bits beyond `avail` are zero.  A codeword of <= 32 bits (all
// counts and nearly all gaps: zeta_3 values < 2^24) costs one CLZ, two shifts for the value and two funnel shifts to
// consume it.  GENERIC: `src` may point to shared memory (staged records) or global memory; otherwise it is global
// and read through the read-only path.  Element 0 of src is stream word j0 (j0 even, so that the 64-bit word halves
// swap as in memory: stream word j = src[(j - j0) ^ 1]).
template <bool GENERIC>
struct BitReaderT {
    const uint32_t* src;
    uint64_t j0;
    uint32_t hi, lo, avail, idx;

    __device__ __forceinline__ uint32_t ld(uint32_t i) const { return GENERIC ? src[i ^ 1u] : __ldg(src + (i ^ 1u)); }
    __device__ __forceinline__ void init(const uint32_t* s, uint64_t j0_, uint64_t p) {
        const uint64_t a = (p >> 6) << 1;  // re-anchor at p's 64-bit word: idx stays small (CGRs beyond 2^37 bits)
        src = s + (a - j0_);
        j0 = a;
        idx = (uint32_t)((p >> 5) - j0);
        const uint32_t off = (uint32_t)(p & 31);
        const uint32_t w0 = ld(idx), w1 = ld(idx + 1);
        hi = __funnelshift_l(w1, w0, off);
        lo = w1 << off;
        avail = 64 - off;
        idx += 2;
    }
    __device__ __forceinline__ uint64_t pos() const { return (j0 + idx) * 32 - avail; }
    __device__ __forceinline__ void refill() {
        if (avail <= 32) {
            const uint32_t w = ld(idx++);
            hi |= __funnelshift_rc(w, 0u, avail);     // w >> avail (0 when avail == 32)
            lo = __funnelshift_lc(0u, w, 32 - avail);  // w << (32 - avail) (0 when avail == 0)
            avail += 32;
        }
    }
    __device__ __forceinline__ void consume(uint32_t L) {  // L <= 32
        hi = __funnelshift_lc(lo, hi, L);
        lo = __funnelshift_lc(0u, lo, L);
        avail -= L;
    }
    // n (1..32) bits; requires avail >= n (true after a refill when n <= 33)
    __device__ __forceinline__ uint32_t take(uint32_t n) {
        const uint32_t v = __funnelshift_rc(hi, 0u, 32 - n);  // hi >> (32 - n), also for n == 32
        consume(n);
        return v;
    }
    template <int K>
    __device__ __forceinline__ uint64_t next() {
        refill();
        const uint32_t z = __clz(hi);
        if (K == 1) {
            if (z < 16) {
                const uint32_t L = 2 * z + 1;
                const uint32_t v = hi >> (32 - L);
                consume(L);
                return v;
            }
        } else {
            const uint32_t h = z + 1, L = h * (K + 1);
            if (L <= 32) {
                const uint32_t v = (hi << h) >> (32 - K * h);
                consume(L);
                return v;
            }
        }
        return next_long<K>(z);
    }
    // Codewords longer than 32 bits (a segment's first residual anchored at u, App. C; far gaps): the prefix is
    // consumed, then the payload is taken in at most two <= 32-bit pieces, refilling in between -- no re-anchoring.
    // Prefixes of 32+ zeros (payloads beyond 64 bits) take the bit-serial path.
    template <int K>
    __device__ __forceinline__ uint64_t next_long(uint32_t z) {
        const uint32_t P = K == 1 ? z + 1 : K * (z + 1);
        if (z >= 32 || P > 64) {
            const Decoded d = decode_at<K, GENERIC>(src, j0, pos());
            init(src, j0, d.end);
            return d.v;
        }
        consume(K == 1 ? z : z + 1);  // K == 1: the payload starts at the leading 1
        refill();
        if (P <= 32) return take(P);
        const uint32_t a = take(P - 32);
        refill();
        return ((uint64_t)a << 32) | take(32);
    }
};
using BitReader = BitReaderT<true>;
using GBitReader = BitReaderT<false>;

// Inverse of the first-gap sign map + 1 (App. C :2101-2106, FORMAT.md R9/R11/R17): code c -> u + delta.
__device__ __forceinline__ uint32_t unmap_first32(uint32_t u, uint64_t c) {
    const uint64_t z = c - 1;
    return (z & 1) ? u - (uint32_t)(z >> 1) : u + (uint32_t)(z >> 1);
}

// ---- warp-cooperative staging of CGR bit ranges into shared memory --------------------------------------------------
// Every lane may ask for one bit range [b, e) (a vertex record, a residual segment).  The ranges are rounded out to
// 16-byte granules (plus 64 bits of slack for the reader's look-ahead), packed back to back into the warp's
// staging buffer in lane order, and copied by the whole warp with coalesced 128-bit loads (LDG.E.128 -> STS.128):
// the misses of all 32 records are in flight together instead of one dependent miss chain per lane.  Ranges that do
// not fit the buffer (or exceed `max_gran` granules) are read from global memory instead.  Returns the reader source
// for the lane's range.
struct StageSlots {
    uint64_t g0[32];    // first granule of each lane's range
    uint32_t excl[32];  // first staging granule of each lane's range
};

template <int CAP>
__device__ __forceinline__ void stage_ranges(uint32_t* __restrict__ buf, uint8_t* __restrict__ owner,
                                             StageSlots& sl, const uint64_t* __restrict__ W, bool want, uint64_t b,
                                             uint64_t e, uint32_t max_gran, const uint32_t*& src, uint64_t& j0) {
    const uint64_t g0 = b >> 7;
    uint32_t ng = want ? (uint32_t)(((e + 64 + 127) >> 7) - g0) : 0u;
    if (ng > max_gran) ng = 0;
    const uint32_t incl = warp_incl_scan(ng), excl = incl - ng;
    const bool fits = ng && incl <= (uint32_t)CAP;
    const uint32_t lane = lane_id();
    if (fits) {
        sl.g0[lane] = g0;
        sl.excl[lane] = excl;
        for (uint32_t k = excl; k < incl; k++) owner[k] = (uint8_t)lane;
    }
    const uint32_t G = __reduce_max_sync(0xffffffffu, fits ? incl : 0u);
    __syncwarp();
    const uint4* __restrict__ W4 = reinterpret_cast<const uint4*>(W);
    uint4* B4 = reinterpret_cast<uint4*>(buf);
    for (uint32_t k = lane; k < G; k += 32) {
        const uint32_t o = owner[k];
        B4[k] = __ldg(W4 + sl.g0[o] + (k - sl.excl[o]));
    }
    __syncwarp();
    if (fits) {
        src = buf + (size_t)excl * 4;
        j0 = g0 * 4;
    } else {
        src = reinterpret_cast<const uint32_t*>(W);
        j0 = 0;
    }
}

__device__ __forceinline__ void add_stats3(unsigned long long* st, uint64_t v, uint64_t a, uint64_t b) {
#pragma unroll
    for (int o = 16; o; o >>= 1) {  // warp reduce (call with the full warp), one reduction per counter per warp
        v += __shfl_xor_sync(0xffffffffu, v, o);
        a += __shfl_xor_sync(0xffffffffu, a, o);
        b += __shfl_xor_sync(0xffffffffu, b, o);
    }
    if (lane_id() == 0) {
        if (v) red_add(st, (unsigned long long)v);
        if (a) red_add(st + 1, (unsigned long long)a);
        if (b) red_add(st + 2, (unsigned long long)b);
    }
}

}  // namespace gcgt_dev

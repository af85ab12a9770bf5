// encode.cpp — host Graph Compression Module: CSR -> CGR (Fig. 3; §3.1 :353-411;
// App. C :2097-2112; §5.2 :1092-1136).  Bit-exact with FORMAT.md R1-R19.
//
// B200-side design: two parallel passes over vertices (OpenMP).  Pass 1 plans every record (intervals, residual
// segments) and sums its bit length; an exclusive prefix gives bit_offsets.  Pass 2 re-plans and writes each
// record into a zeroed array of 64-bit words in stream order (bit i of the stream = bit 63-(i%64) of word i/64),
// OR-ing the two words a record may share with its neighbours atomically.  A final byte swap turns the words into
// the canonical MSB-first byte stream in place.  Zero bits are never written (the array starts zeroed), so unary
// prefixes and segment padding cost nothing.
#include <omp.h>
#include <stdio.h>
#include <string.h>

#include <algorithm>
#include <atomic>
#include <memory>
#include <new>

#include "internal.h"

namespace {

inline int bitlen(uint64_t x) { return x ? 64 - __builtin_clzll(x) : 0; }

// Code length of VLC_k(x) (App. B; FORMAT.md R3/R4).
inline uint32_t code_len(uint32_t k, uint64_t x) {
    const int b = bitlen(x);
    if (k == 1) return (uint32_t)(2 * b - 1);
    const int h = (b + (int)k - 1) / (int)k;
    return (uint32_t)(h * ((int)k + 1));
}

// Sign map of the first gap (App. C :2101-2106), then "+1" (:2111).
inline uint64_t first_code(int64_t delta) { return (delta >= 0 ? 2 * (uint64_t)delta : 2 * (uint64_t)(-delta) + 1) + 1; }

struct Interval { uint32_t start, len; };

// Per-thread scratch for one vertex's plan.
struct Plan {
    std::vector<Interval> itv;
    std::vector<uint32_t> res;
    std::vector<uint32_t> seg_cnt;  // residuals per segment (segmented format only)
    uint64_t bits = 0;
};

// Splits row u into intervals / residuals (R7), packs residual segments (R18) and returns the record length.
gcgt_status plan_vertex(uint64_t u, const uint32_t* row, uint64_t deg, const gcgt_params& P, Plan& pl) {
    const uint32_t k = P.zeta_k, ml = P.min_interval_len;
    pl.itv.clear();
    pl.res.clear();
    pl.seg_cnt.clear();
    uint64_t i = 0;
    while (i < deg) {
        uint64_t j = i + 1;
        while (j < deg && row[j] == row[j - 1] + 1) j++;
        if (ml && j - i >= ml) pl.itv.push_back({row[i], (uint32_t)(j - i)});
        else pl.res.insert(pl.res.end(), row + i, row + j);
        i = j;
    }
    uint64_t L = 0;
    if (P.residual_segment_len == 0) L += code_len(k, deg + 1);
    L += code_len(k, pl.itv.size() + 1);
    for (size_t t = 0; t < pl.itv.size(); t++) {
        const Interval& iv = pl.itv[t];
        L += t == 0 ? code_len(k, first_code((int64_t)iv.start - (int64_t)u))
                    : code_len(k, (uint64_t)iv.start - (pl.itv[t - 1].start + pl.itv[t - 1].len - 1));
        L += code_len(k, iv.len - ml + 1);
    }
    const uint64_t R = pl.res.size();
    if (P.residual_segment_len == 0) {
        for (uint64_t t = 0; t < R; t++)
            L += t == 0 ? code_len(k, first_code((int64_t)pl.res[0] - (int64_t)u))
                        : code_len(k, (uint64_t)(pl.res[t] - pl.res[t - 1]));
        pl.bits = L;
        return GCGT_OK;
    }
    // Segmented: greedy packing with the last-segment rule (R16-R19).
    const uint64_t segBits = 8ull * P.residual_segment_len;
    uint64_t gap_tail = 0;  // sum of gap-code lengths of res[p+1 .. R-1] for the current start p
    for (uint64_t t = 1; t < R; t++) gap_tail += code_len(k, (uint64_t)(pl.res[t] - pl.res[t - 1]));
    uint64_t p = 0, seg_bits_total = 0;
    while (p < R) {
        const uint64_t head = code_len(k, first_code((int64_t)pl.res[p] - (int64_t)u));
        const uint64_t whole = code_len(k, R - p + 1) + head + gap_tail;
        if (whole <= 2 * segBits) {  // last segment, unpadded
            pl.seg_cnt.push_back((uint32_t)(R - p));
            seg_bits_total += whole;
            break;
        }
        uint64_t c = 1, body_gaps = 0;
        if (code_len(k, 2) + head > segBits) return gcgt_internal::fail(GCGT_ESEGLEN, "residual segment too short");
        while (p + c < R) {
            const uint64_t g = code_len(k, (uint64_t)(pl.res[p + c] - pl.res[p + c - 1]));
            if (code_len(k, c + 2) + head + body_gaps + g > segBits) break;
            body_gaps += g;
            c++;
        }
        // advance: drop the gaps inside this segment and the (re-anchored) gap into the next one
        gap_tail -= body_gaps;
        if (p + c < R) gap_tail -= code_len(k, (uint64_t)(pl.res[p + c] - pl.res[p + c - 1]));
        pl.seg_cnt.push_back((uint32_t)c);
        seg_bits_total += segBits;
        p += c;
    }
    L += code_len(k, pl.seg_cnt.size() + 1) + seg_bits_total;
    pl.bits = L;
    return GCGT_OK;
}

// Stream writer over the shared word array; words [lo_w, hi_w] are the record's first/last (possibly shared).
struct Writer {
    uint64_t* W;
    uint64_t pos;
    uint64_t lo_w, hi_w;
    inline void or_word(uint64_t i, uint64_t v) {
        if (!v) return;
        if (i == lo_w || i == hi_w) __atomic_fetch_or(&W[i], v, __ATOMIC_RELAXED);
        else W[i] |= v;
    }
    inline void put(uint64_t x, uint32_t nb) {  // low nb bits of x (nb <= 64) at pos
        if (nb == 0) return;
        const uint64_t i = pos >> 6;
        const uint32_t o = (uint32_t)(pos & 63);
        if (nb < 64) x &= (1ull << nb) - 1;
        if (o + nb <= 64) {
            or_word(i, x << (64 - o - nb));
        } else {
            const uint32_t spill = o + nb - 64;  // bits that go to word i+1
            or_word(i, x >> spill);
            or_word(i + 1, x << (64 - spill));
        }
        pos += nb;
    }
    inline void code(uint32_t k, uint64_t x) {
        const int b = bitlen(x);
        if (k == 1) {  // (b-1) zeros, then b bits
            pos += (uint64_t)(b - 1);
            put(x, (uint32_t)b);
        } else {       // (h-1) zeros, '1', x in h*k bits
            const int h = (b + (int)k - 1) / (int)k;
            pos += (uint64_t)(h - 1);
            put(1, 1);
            const uint32_t w = (uint32_t)(h * (int)k);
            if (w > 64) pos += w - 64;
            put(x, w > 64 ? 64 : w);
        }
    }
};

void write_vertex(uint64_t u, const Plan& pl, uint64_t deg, const gcgt_params& P, Writer& w) {
    const uint32_t k = P.zeta_k, ml = P.min_interval_len;
    if (P.residual_segment_len == 0) w.code(k, deg + 1);
    w.code(k, pl.itv.size() + 1);
    for (size_t t = 0; t < pl.itv.size(); t++) {
        const Interval& iv = pl.itv[t];
        w.code(k, t == 0 ? first_code((int64_t)iv.start - (int64_t)u)
                         : (uint64_t)iv.start - (pl.itv[t - 1].start + pl.itv[t - 1].len - 1));
        w.code(k, iv.len - ml + 1);
    }
    const uint64_t R = pl.res.size();
    if (P.residual_segment_len == 0) {
        for (uint64_t t = 0; t < R; t++)
            w.code(k, t == 0 ? first_code((int64_t)pl.res[0] - (int64_t)u) : (uint64_t)(pl.res[t] - pl.res[t - 1]));
        return;
    }
    const uint64_t segBits = 8ull * P.residual_segment_len;
    w.code(k, pl.seg_cnt.size() + 1);
    const uint64_t base = w.pos;
    uint64_t p = 0;
    for (size_t s = 0; s < pl.seg_cnt.size(); s++) {
        w.pos = base + s * segBits;
        const uint32_t c = pl.seg_cnt[s];
        w.code(k, (uint64_t)c + 1);
        w.code(k, first_code((int64_t)pl.res[p] - (int64_t)u));
        for (uint32_t t = 1; t < c; t++) w.code(k, (uint64_t)(pl.res[p + t] - pl.res[p + t - 1]));
        p += c;
    }
}

}  // namespace

// Encodes rows 0..csr->n-1 as the records of vertices first .. first + csr->n - 1 of a graph of n_total vertices.
static gcgt_status encode_rows(const gcgt_csr* csr, uint64_t first, uint64_t n_total, const gcgt_params* params,
                               gcgt_cgr** out) {
    using gcgt_internal::fail;
    gcgt_internal::clear_error();
    if (!csr || !params || !out) return fail(GCGT_EINVAL, "null argument");
    const gcgt_params P = *params;
    if (P.zeta_k < 1 || P.zeta_k > 5) return fail(GCGT_EINVAL, "zeta_k must be 1..5");
    if (P.min_interval_len == 1) return fail(GCGT_EINVAL, "min_interval_len must be 0 or >= 2");
    const uint64_t n = csr->n;
    if (n_total > 0xFFFFFFFFull || first + n > n_total) return fail(GCGT_EINVAL, "n must fit in uint32");
    if (n && (!csr->row_offsets || (!csr->cols && csr->row_offsets[n] > 0)))
        return fail(GCGT_EINVAL, "null CSR arrays");
    const uint64_t* ro = csr->row_offsets;
    const uint32_t* cols = csr->cols;
    // validate (R6) before any allocation
    int bad = 0;  // 1 EINVAL, 2 ERANGE, 3 EUNSORTED
    if (n && ro[0] != 0) bad = 1;
#pragma omp parallel for schedule(dynamic, 4096) reduction(max : bad)
    for (int64_t u = 0; u < (int64_t)n; u++) {
        if (ro[u + 1] < ro[u]) { bad = std::max(bad, 1); continue; }
        for (uint64_t e = ro[u]; e < ro[u + 1]; e++) {
            if (cols[e] >= n_total) bad = std::max(bad, 2);
            else if (e > ro[u] && cols[e] <= cols[e - 1]) bad = std::max(bad, 3);
        }
    }
    if (bad == 1) return fail(GCGT_EINVAL, "row_offsets not non-decreasing from 0");
    if (bad == 2) return fail(GCGT_ERANGE, "column id >= n");
    if (bad == 3) return fail(GCGT_EUNSORTED, "row not strictly increasing");

    std::unique_ptr<gcgt_cgr> g;
    try {
        g.reset(new gcgt_cgr());
        g->n = n;
        g->base = first;
        g->n_total = n_total;
        g->params = P;
        g->bit_offsets.assign(n + 1, 0);
    } catch (...) {
        return fail(GCGT_ENOMEM, "host allocation failed");
    }
    // pass 1: lengths
    std::atomic<int> err{GCGT_OK};
#pragma omp parallel
    {
        Plan pl;
#pragma omp for schedule(dynamic, 1024)
        for (int64_t u = 0; u < (int64_t)n; u++) {
            if (err.load(std::memory_order_relaxed) != GCGT_OK) continue;
            gcgt_status st = plan_vertex(first + (uint64_t)u, cols + ro[u], ro[u + 1] - ro[u], P, pl);
            if (st != GCGT_OK) { err.store(st); continue; }
            g->bit_offsets[u + 1] = pl.bits;
        }
    }
    if (err.load() != GCGT_OK) return fail((gcgt_status)err.load(), "residual segment too short (FORMAT.md R19)");
    for (uint64_t u = 0; u < n; u++) g->bit_offsets[u + 1] += g->bit_offsets[u];
    g->nbits = g->bit_offsets[n];
    const uint64_t nwords = (g->nbits + 63) / 64 + 2;
    try {
        g->words.assign(nwords, 0);
    } catch (...) {
        return fail(GCGT_ENOMEM, "host allocation failed");
    }
    // pass 2: write
#pragma omp parallel
    {
        Plan pl;
#pragma omp for schedule(dynamic, 1024)
        for (int64_t u = 0; u < (int64_t)n; u++) {
            const uint64_t b0 = g->bit_offsets[u], b1 = g->bit_offsets[u + 1];
            if (b1 == b0) continue;
            plan_vertex(first + (uint64_t)u, cols + ro[u], ro[u + 1] - ro[u], P, pl);
            Writer w{g->words.data(), b0, b0 >> 6, (b1 - 1) >> 6};
            write_vertex(first + (uint64_t)u, pl, ro[u + 1] - ro[u], P, w);
        }
    }
    // words (stream order) -> canonical bytes in memory order
#pragma omp parallel for schedule(static)
    for (int64_t i = 0; i < (int64_t)nwords; i++) g->words[i] = __builtin_bswap64(g->words[i]);
    *out = g.release();
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_encode(const gcgt_csr* csr, const gcgt_params* params, gcgt_cgr** out) {
    return encode_rows(csr, 0, csr ? csr->n : 0, params, out);
}

extern "C" gcgt_status gcgt_encode_slice(const gcgt_csr* rows, uint64_t first, uint64_t n_total,
                                         const gcgt_params* params, gcgt_cgr** out) {
    return encode_rows(rows, first, n_total, params, out);
}

// Concatenation of consecutive vertex-range slices (R2: records are concatenated in vertex order, so the slices'
// bit streams are appended at the running bit total and their offsets shifted by it).
extern "C" gcgt_status gcgt_cgr_concat(const gcgt_cgr* const* parts, uint32_t k, gcgt_cgr** out) {
    using gcgt_internal::fail;
    gcgt_internal::clear_error();
    if (!parts || !out || k == 0) return fail(GCGT_EINVAL, "null argument");
    for (uint32_t i = 0; i < k; i++) {
        if (!parts[i]) return fail(GCGT_EINVAL, "null part");
        const gcgt_params& a = parts[i]->params;
        const gcgt_params& b = parts[0]->params;
        if (a.zeta_k != b.zeta_k || a.min_interval_len != b.min_interval_len ||
            a.residual_segment_len != b.residual_segment_len || parts[i]->n_total != parts[0]->n_total)
            return fail(GCGT_EINVAL, "parts differ in parameters or graph size");
        if (i && parts[i]->base != parts[i - 1]->base + parts[i - 1]->n)
            return fail(GCGT_EINVAL, "parts are not consecutive vertex ranges");
    }
    std::unique_ptr<gcgt_cgr> g;
    std::vector<uint64_t> start(k + 1, 0);
    for (uint32_t i = 0; i < k; i++) start[i + 1] = start[i] + parts[i]->nbits;
    uint64_t n = 0;
    for (uint32_t i = 0; i < k; i++) n += parts[i]->n;
    try {
        g.reset(new gcgt_cgr());
        g->n = n;
        g->base = parts[0]->base;
        g->n_total = parts[0]->n_total;
        g->params = parts[0]->params;
        g->nbits = start[k];
        g->bit_offsets.resize(n + 1);
        g->words.assign((g->nbits + 63) / 64 + 2, 0);
    } catch (...) {
        return fail(GCGT_ENOMEM, "host allocation failed");
    }
    uint64_t v0 = 0;
    for (uint32_t i = 0; i < k; i++) {
        const gcgt_cgr* p = parts[i];
        const uint64_t sh = start[i];
#pragma omp parallel for schedule(static)
        for (int64_t u = 0; u < (int64_t)p->n; u++) g->bit_offsets[v0 + u] = p->bit_offsets[u] + sh;
        v0 += p->n;
        // append the part's bits at bit `sh`: stream words (byte-swapped canonical words) shifted right by sh % 64;
        // the first word is shared with the previous part (OR), the others are written whole
        const uint64_t nw = (p->nbits + 63) / 64, w0 = sh / 64, s = sh % 64;
        uint64_t* dst = g->words.data();
        const uint64_t* src = p->words.data();
        auto sw = [&](uint64_t j) { return j < nw ? __builtin_bswap64(src[j]) : 0ull; };
        if (nw) {
            const uint64_t first = sw(0) >> s;
            dst[w0] = __builtin_bswap64(__builtin_bswap64(dst[w0]) | first);
#pragma omp parallel for schedule(static)
            for (int64_t j = 1; j <= (int64_t)nw; j++) {
                const uint64_t v = (s ? sw(j - 1) << (64 - s) : 0ull) | (sw(j) >> s);
                if (w0 + j < g->words.size()) dst[w0 + j] = __builtin_bswap64(v);
            }
        }
    }
    g->bit_offsets[n] = g->nbits;
    *out = g.release();
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_cgr_slice_info(const gcgt_cgr* c, uint64_t* base, uint64_t* n_total) {
    gcgt_internal::clear_error();
    if (!c) return gcgt_internal::fail(GCGT_EINVAL, "null cgr");
    if (base) *base = c->base;
    if (n_total) *n_total = c->n_total;
    return GCGT_OK;
}

// Transpose on the host (parallel counting sort by target), then the same encoder.
extern "C" gcgt_status gcgt_encode_transpose(const gcgt_csr* csr, const gcgt_params* params, gcgt_cgr** out) {
    using gcgt_internal::fail;
    gcgt_internal::clear_error();
    if (!csr || !params || !out) return fail(GCGT_EINVAL, "null argument");
    const uint64_t n = csr->n;
    const uint64_t m = n ? csr->row_offsets[n] : 0;
    const uint64_t* ro = csr->row_offsets;
    const uint32_t* cols = csr->cols;
    for (uint64_t e = 0; e < m; e++)
        if (cols[e] >= n) return fail(GCGT_ERANGE, "column id >= n");
    std::vector<uint64_t> tro;
    std::vector<uint32_t> tco;
    try {
        tro.assign(n + 1, 0);
        tco.resize(m);
    } catch (...) {
        return fail(GCGT_ENOMEM, "host allocation failed");
    }
    for (uint64_t e = 0; e < m; e++) tro[cols[e] + 1]++;
    for (uint64_t v = 0; v < n; v++) tro[v + 1] += tro[v];
    // rows are emitted in increasing source order, so every transposed row comes out sorted
    std::vector<uint64_t> pos(tro.begin(), tro.end() - (n ? 1 : 0));
    for (uint64_t u = 0; u < n; u++)
        for (uint64_t e = ro[u]; e < ro[u + 1]; e++) tco[pos[cols[e]]++] = (uint32_t)u;
    const gcgt_csr t{n, tro.data(), tco.data()};
    return gcgt_encode(&t, params, out);
}

extern "C" gcgt_status gcgt_cgr_view(const gcgt_cgr* c, const uint8_t** bytes, uint64_t* nbits,
                                     const uint64_t** bit_offsets, uint64_t* n, gcgt_params* params) {
    gcgt_internal::clear_error();
    if (!c) return gcgt_internal::fail(GCGT_EINVAL, "null cgr");
    if (bytes) *bytes = (const uint8_t*)c->words.data();
    if (nbits) *nbits = c->nbits;
    if (bit_offsets) *bit_offsets = c->bit_offsets.data();
    if (n) *n = c->n;
    if (params) *params = c->params;
    return GCGT_OK;
}

static gcgt_status check_params(const gcgt_params& P) {
    if (P.zeta_k < 1 || P.zeta_k > 5 || P.min_interval_len == 1)
        return gcgt_internal::fail(GCGT_EFORMAT, "bad CGR parameters");
    return GCGT_OK;
}

// Shared validation of an externally supplied CGR (gcgt_cgr_from_arrays, gcgt_cgr_open): 32-bit vertex ids, bit
// offsets starting at 0, non-decreasing, ending at nbits.  Corrupt tables would otherwise reach the device decoders.
static gcgt_status check_offsets(uint64_t n, uint64_t nbits, const uint64_t* bit_offsets) {
    using gcgt_internal::fail;
    if (n >= 0xFFFFFFFFull) return fail(GCGT_EFORMAT, "n must fit 32-bit vertex ids");
    if (bit_offsets[0] != 0 || bit_offsets[n] != nbits) return fail(GCGT_EFORMAT, "bit_offsets[0] != 0 or [n] != nbits");
    for (uint64_t u = 0; u < n; u++)
        if (bit_offsets[u + 1] < bit_offsets[u]) return fail(GCGT_EFORMAT, "bit_offsets decreasing");
    return GCGT_OK;
}

extern "C" gcgt_status gcgt_cgr_from_arrays(uint64_t n, const uint8_t* bytes, uint64_t nbits,
                                            const uint64_t* bit_offsets, const gcgt_params* params,
                                            gcgt_cgr** out) {
    using gcgt_internal::fail;
    gcgt_internal::clear_error();
    if (!bit_offsets || !params || !out || (nbits && !bytes)) return fail(GCGT_EINVAL, "null argument");
    if (check_params(*params) != GCGT_OK) return GCGT_EFORMAT;
    if (gcgt_status st = check_offsets(n, nbits, bit_offsets)) return st;
    try {
        std::unique_ptr<gcgt_cgr> g(new gcgt_cgr());
        g->n = n;
        g->n_total = n;
        g->nbits = nbits;
        g->params = *params;
        g->bit_offsets.assign(bit_offsets, bit_offsets + n + 1);
        g->words.assign((nbits + 63) / 64 + 2, 0);
        memcpy(g->words.data(), bytes, (nbits + 7) / 8);
        *out = g.release();
    } catch (...) {
        return fail(GCGT_ENOMEM, "host allocation failed");
    }
    return GCGT_OK;
}

// File layout: "GCGTCGR2" | n u64 | nbits u64 | min_interval_len, residual_segment_len, zeta_k, 0 (u32 x4) |
// base u64 | n_total u64 | bit_offsets u64[n+1] | bytes[ceil(nbits/8)].  ("GCGTCGR1" files: no base / n_total.)
extern "C" gcgt_status gcgt_cgr_save(const gcgt_cgr* c, const char* path) {
    using gcgt_internal::fail;
    gcgt_internal::clear_error();
    if (!c || !path) return fail(GCGT_EINVAL, "null argument");
    FILE* f = fopen(path, "wb");
    if (!f) return fail(GCGT_EINVAL, std::string("cannot open ") + path);
    const uint32_t pr[4] = {c->params.min_interval_len, c->params.residual_segment_len, c->params.zeta_k, 0};
    bool ok = fwrite("GCGTCGR2", 1, 8, f) == 8 && fwrite(&c->n, 8, 1, f) == 1 && fwrite(&c->nbits, 8, 1, f) == 1 &&
              fwrite(pr, 4, 4, f) == 4 && fwrite(&c->base, 8, 1, f) == 1 && fwrite(&c->n_total, 8, 1, f) == 1 &&
              fwrite(c->bit_offsets.data(), 8, c->n + 1, f) == c->n + 1 &&
              fwrite(c->words.data(), 1, c->nbytes(), f) == c->nbytes();
    ok = (fclose(f) == 0) && ok;
    return ok ? GCGT_OK : fail(GCGT_EINVAL, "write failed");
}

extern "C" gcgt_status gcgt_cgr_open(const char* path, gcgt_cgr** out) {
    using gcgt_internal::fail;
    gcgt_internal::clear_error();
    if (!path || !out) return fail(GCGT_EINVAL, "null argument");
    FILE* f = fopen(path, "rb");
    if (!f) return fail(GCGT_EINVAL, std::string("cannot open ") + path);
    char magic[8];
    uint64_t n = 0, nbits = 0, base = 0, n_total = 0;
    uint32_t pr[4];
    gcgt_status st = GCGT_OK;
    std::unique_ptr<gcgt_cgr> g;
    bool v2 = false;
    if (fread(magic, 1, 8, f) != 8 || (memcmp(magic, "GCGTCGR1", 8) && !(v2 = !memcmp(magic, "GCGTCGR2", 8))) ||
        fread(&n, 8, 1, f) != 1 || fread(&nbits, 8, 1, f) != 1 || fread(pr, 4, 4, f) != 4 ||
        (v2 && (fread(&base, 8, 1, f) != 1 || fread(&n_total, 8, 1, f) != 1))) {
        st = fail(GCGT_EFORMAT, "bad CGR file header");
    } else if (!v2 && (n_total = n, false)) {
    } else if (n >= 0xFFFFFFFFull || nbits / 8 > (1ull << 42) || n_total >= 0xFFFFFFFFull || base + n > n_total) {
        st = fail(GCGT_EFORMAT, "CGR file header out of range");
    } else {
        try {
            g.reset(new gcgt_cgr());
            g->n = n;
            g->base = base;
            g->n_total = n_total;
            g->nbits = nbits;
            g->params = {pr[0], pr[1], pr[2]};
            g->bit_offsets.resize(n + 1);
            g->words.assign((nbits + 63) / 64 + 2, 0);
        } catch (...) {
            st = fail(GCGT_ENOMEM, "host allocation failed");
        }
        if (st == GCGT_OK && (fread(g->bit_offsets.data(), 8, n + 1, f) != n + 1 ||
                              fread(g->words.data(), 1, g->nbytes(), f) != g->nbytes()))
            st = fail(GCGT_EFORMAT, "truncated CGR file");
        if (st == GCGT_OK && check_params(g->params) != GCGT_OK) st = fail(GCGT_EFORMAT, "inconsistent CGR file");
        if (st == GCGT_OK) st = check_offsets(n, nbits, g->bit_offsets.data());
    }
    fclose(f);
    if (st == GCGT_OK) *out = g.release();
    return st;
}

extern "C" void gcgt_cgr_free(gcgt_cgr* c) {
    if (!c) return;
    gcgt_internal::release_tables(c);
    delete c;
}

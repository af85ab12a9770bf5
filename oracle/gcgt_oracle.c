/*
 * gcgt_oracle.c — plain, slow, obviously-correct CPU oracle for GCGT (Sha, Li, Tan, SIGMOD '19).
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference
 * legs may load this library.  It shares no code, header, table or helper with the product path
 * (paper_conf_sigmod_shalt19_b200/csrc/), and the product never loads it.
 *
 * Every function cites the passage it follows: PAPER.md:<line> (+ section / algorithm / figure) and the
 * FORMAT.md rule number.  The format readings are listed in DESIGN.md §3.
 *
 * Pins (tests/test_oracle_*.py, -m "not gpu"):
 *   orc_vlc_*            Table 3 (24 codewords), round trip, Fig. 5 vals/poss
 *   orc_encode (illustr) Fig. 2 (55 bits, exact)
 *   orc_encode (canon.)  derived worked examples (FORMAT.md), round trip, bit-length identity, layout invariants
 *   orc_alg4_trace       Fig. 5 round-by-round trace, Lemma 5.2 round bound
 *   orc_bfs / _cgr       Fig. 1 levels, Bellman-Ford fixpoint on random small graphs
 *   orc_cc               brute-force reachability, Fig. 1
 *   orc_bc               brute-force pair counting (definition), closed forms (path, star, cycle, complete)
 * All functions are pinned; none is "parity unpinned".
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

enum { ORC_OK = 0, ORC_EINVAL = -1, ORC_EUNSORTED = -2, ORC_ERANGE = -3, ORC_ESEGLEN = -4, ORC_ENOMEM = -5,
       ORC_EFORMAT = -8 };

/* ------------------------------------------------------------------------------------------------------------ */
/* Bit stream, MSB-first (FORMAT.md R1).                                                                          */
/* ------------------------------------------------------------------------------------------------------------ */
typedef struct { uint8_t *buf; uint64_t nbits; uint64_t capbytes; int oom; } bitbuf;

static void bb_put(bitbuf *b, int bit) {
    if ((b->nbits >> 3) >= b->capbytes) {
        uint64_t nc = b->capbytes ? 2 * b->capbytes : 64;
        uint8_t *nb = (uint8_t *)realloc(b->buf, nc);
        if (!nb) { b->oom = 1; return; }
        memset(nb + b->capbytes, 0, nc - b->capbytes);
        b->buf = nb; b->capbytes = nc;
    }
    if (bit) b->buf[b->nbits >> 3] |= (uint8_t)(0x80u >> (b->nbits & 7));
    b->nbits++;
}

static int bit_at(const uint8_t *bytes, uint64_t i) { return (bytes[i >> 3] >> (7 - (i & 7))) & 1; }

static int nbits_of(uint64_t x) { int b = 0; while (x) { b++; x >>= 1; } return b; }

/* ------------------------------------------------------------------------------------------------------------ */
/* VLC codes (App. B, Table 3 :1854-1864; FORMAT.md R3, R4).                                   */
/* ------------------------------------------------------------------------------------------------------------ */

/* Length in bits of VLC_k(x), x >= 1. */
uint64_t orc_vlc_len(int k, uint64_t x) {
    int b = nbits_of(x);
    if (k == 1) return (uint64_t)(2 * b - 1);            /* R3: (b-1) zeros + b bits            */
    int h = (b + k - 1) / k;                             /* R4: h = ceil(b/k)                    */
    return (uint64_t)(h + h * k);                        /*     (h-1) zeros + '1' + h*k bits     */
}

static void vlc_put(bitbuf *bb, int k, uint64_t x) {
    int b = nbits_of(x);
    if (k == 1) {                                        /* R3 */
        for (int i = 0; i < b - 1; i++) bb_put(bb, 0);
        for (int i = b - 1; i >= 0; i--) bb_put(bb, (int)((x >> i) & 1));
    } else {                                             /* R4 */
        int h = (b + k - 1) / k;
        for (int i = 0; i < h - 1; i++) bb_put(bb, 0);
        bb_put(bb, 1);
        for (int i = h * k - 1; i >= 0; i--) bb_put(bb, i < 64 ? (int)((x >> i) & 1) : 0);
    }
}

/* Writes VLC_k(x) as a '0'/'1' string (for the Table 3 pin).  Returns its length, or -1. */
int orc_vlc_string(int k, uint64_t x, char *out, int cap) {
    if (x == 0 || k < 1 || k > 5) return -1;
    bitbuf bb = {0};
    vlc_put(&bb, k, x);
    if (bb.oom || (int)bb.nbits + 1 > cap) { free(bb.buf); return -1; }
    for (uint64_t i = 0; i < bb.nbits; i++) out[i] = (char)('0' + bit_at(bb.buf, i));
    out[bb.nbits] = 0;
    int n = (int)bb.nbits;
    free(bb.buf);
    return n;
}

/* Decodes one codeword starting at stream bit *pos (the paper's decodeNum, Alg. 1 l.6, :581-584).
 * Returns 0 and advances *pos, or -1 if the codeword runs past nbits or is longer than 64 payload bits. */
int orc_vlc_read(int k, const uint8_t *bytes, uint64_t nbits, uint64_t *pos, uint64_t *val) {
    uint64_t p = *pos, zeros = 0;
    while (p < nbits && !bit_at(bytes, p)) { zeros++; p++; }
    if (p >= nbits) return -1;
    uint64_t payload;
    if (k == 1) {
        payload = zeros + 1;                              /* R3: the leading 1 is part of x */
    } else {
        p++;                                              /* R4: skip the terminating 1 of the unary part */
        payload = (zeros + 1) * (uint64_t)k;
    }
    if (p + payload > nbits) return -1;
    uint64_t x = 0;
    for (uint64_t i = 0; i < payload; i++) {
        if (x >> 63) return -1;                           /* value does not fit in 64 bits */
        x = (x << 1) | (uint64_t)bit_at(bytes, p + i);
    }
    *pos = p + payload;
    *val = x;
    return 0;
}

/* ------------------------------------------------------------------------------------------------------------ */
/* Encoder (§3.1 :353-411, App. C :2097-2112, §5.2 :1092-1136; FORMAT.md R6-R19).                                 */
/* ------------------------------------------------------------------------------------------------------------ */
static uint64_t sm(int64_t x) { return x >= 0 ? (uint64_t)(2 * x) : (uint64_t)(2 * (-x) + 1); }  /* App. C :2101-2106 */

/* Bit length of a segment body holding residuals r[0..c-1] of vertex u (R17). */
static uint64_t seg_body_len(int k, uint64_t u, const uint32_t *r, uint64_t c) {
    uint64_t L = orc_vlc_len(k, c + 1);
    L += orc_vlc_len(k, sm((int64_t)r[0] - (int64_t)u) + 1);
    for (uint64_t i = 1; i < c; i++) L += orc_vlc_len(k, (uint64_t)(r[i] - r[i - 1]));
    return L;
}

static void seg_body_put(bitbuf *bb, int k, uint64_t u, const uint32_t *r, uint64_t c) {
    vlc_put(bb, k, c + 1);
    vlc_put(bb, k, sm((int64_t)r[0] - (int64_t)u) + 1);
    for (uint64_t i = 1; i < c; i++) vlc_put(bb, k, (uint64_t)(r[i] - r[i - 1]));
}

/* Encodes the record of vertex u (list adj[0..deg-1]) onto bb.  illustrative != 0 selects Fig. 2's raw mode. */
static int encode_vertex(bitbuf *bb, uint64_t u, const uint32_t *adj, uint64_t deg, uint32_t minLen,
                         uint32_t segLen, int k, int illustrative, uint32_t *itv_start, uint32_t *itv_len,
                         uint32_t *res) {
    /* R7: maximal runs of consecutive ids; runs of length >= minLen become intervals, the rest residuals. */
    uint64_t nitv = 0, nres = 0, i = 0;
    while (i < deg) {
        uint64_t j = i + 1;
        while (j < deg && adj[j] == adj[j - 1] + 1) j++;
        uint64_t run = j - i;
        if (minLen != 0 && run >= minLen) {
            itv_start[nitv] = adj[i]; itv_len[nitv] = (uint32_t)run; nitv++;
        } else {
            for (uint64_t t = i; t < j; t++) res[nres++] = adj[t];
        }
        i = j;
    }
    if (illustrative) {
        /* Fig. 2 (:387-399): degNum, itvNum, (gap,len)*, residual gaps; no App. C shifts.  Zero values cannot be
         * coded (the VLC has no code for 0, App. C :2111), so they are an error in this mode. */
        if (deg == 0) return ORC_EINVAL;
        vlc_put(bb, 1, deg);
        if (nitv == 0) return ORC_EINVAL;
        vlc_put(bb, 1, nitv);
        for (uint64_t t = 0; t < nitv; t++) {
            uint64_t g = t == 0 ? sm((int64_t)itv_start[0] - (int64_t)u)
                                : (uint64_t)(itv_start[t] - (itv_start[t - 1] + itv_len[t - 1] - 1));
            if (g == 0) return ORC_EINVAL;
            vlc_put(bb, 1, g);
            vlc_put(bb, 1, itv_len[t]);
        }
        for (uint64_t t = 0; t < nres; t++) {
            uint64_t g = t == 0 ? sm((int64_t)res[0] - (int64_t)u) : (uint64_t)(res[t] - res[t - 1]);
            if (g == 0) return ORC_EINVAL;
            vlc_put(bb, 1, g);
        }
        return ORC_OK;
    }
    if (segLen == 0) vlc_put(bb, k, deg + 1);                                  /* R8: degNum (+1)        */
    vlc_put(bb, k, nitv + 1);                                                  /* R8/R14: itvNum (+1)    */
    for (uint64_t t = 0; t < nitv; t++) {
        if (t == 0) vlc_put(bb, k, sm((int64_t)itv_start[0] - (int64_t)u) + 1);              /* R9  */
        else vlc_put(bb, k, (uint64_t)(itv_start[t] - (itv_start[t - 1] + itv_len[t - 1] - 1)));  /* R10 */
        vlc_put(bb, k, (uint64_t)(itv_len[t] - minLen + 1));                                 /* R8 len shift */
    }
    if (segLen == 0) {
        for (uint64_t t = 0; t < nres; t++) {
            if (t == 0) vlc_put(bb, k, sm((int64_t)res[0] - (int64_t)u) + 1);  /* R11 */
            else vlc_put(bb, k, (uint64_t)(res[t] - res[t - 1]));               /* R12 */
        }
        return ORC_OK;
    }
    /* R18 packing: first decide every segment, then write segNum and the segments (R14, R16).
     * L(rest from i) = len(VLC(cnt+1)) + len(VLC(sm(r_i - u)+1)) + sum of the gap codes after r_i; the gap-code
     * sum is a suffix sum G[i] so that each test is O(1) (hub lists have millions of residuals). */
    uint64_t segBits = 8ull * segLen;
    uint64_t nseg = 0, placed = 0;
    uint64_t *segcnt = (uint64_t *)malloc(sizeof(uint64_t) * (nres + 1));
    uint64_t *G = (uint64_t *)malloc(sizeof(uint64_t) * (nres + 1));
    if (!segcnt || !G) { free(segcnt); free(G); return ORC_ENOMEM; }
    if (nres) G[nres - 1] = 0;
    for (uint64_t t = nres - 1; nres && t-- > 0;) G[t] = G[t + 1] + orc_vlc_len(k, (uint64_t)(res[t + 1] - res[t]));
    while (placed < nres) {
        uint64_t rest = nres - placed;
        uint64_t Lrest = orc_vlc_len(k, rest + 1) + orc_vlc_len(k, sm((int64_t)res[placed] - (int64_t)u) + 1) +
                         G[placed];
        if (Lrest <= 2 * segBits) {                                    /* last segment, unpadded */
            segcnt[nseg++] = rest; placed = nres; break;
        }
        uint64_t c = 0;                                                /* longest prefix fitting segBits */
        while (c + 1 <= rest && seg_body_len(k, u, res + placed, c + 1) <= segBits) c++;
        if (c == 0) { free(segcnt); free(G); return ORC_ESEGLEN; }     /* R19 */
        segcnt[nseg++] = c; placed += c;
    }
    free(G);
    vlc_put(bb, k, nseg + 1);                                          /* R14: segNum (+1) */
    placed = 0;
    for (uint64_t s = 0; s < nseg; s++) {
        uint64_t start = bb->nbits;
        seg_body_put(bb, k, u, res + placed, segcnt[s]);               /* R17 */
        placed += segcnt[s];
        if (s + 1 < nseg) while (bb->nbits - start < segBits) bb_put(bb, 0);   /* R16 blank padding */
    }
    free(segcnt);
    return ORC_OK;
}

/* CSR -> CGR (Fig. 3 :438-454 "Graph Compression Module").  On success *bytes_out is malloc'ed (caller frees with
 * orc_free), *nbits_out = total bits, bit_offsets[0..n] filled (R2). */
int orc_encode(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, uint32_t minLen, uint32_t segLen,
               uint32_t k, uint8_t **bytes_out, uint64_t *nbits_out, uint64_t *bit_offsets) {
    if (minLen == 1 || k < 1 || k > 5) return ORC_EINVAL;
    uint64_t maxdeg = 0;
    for (uint64_t u = 0; u < n; u++) {                                  /* R6: validate every row */
        if (rowoff[u + 1] < rowoff[u]) return ORC_EINVAL;
        uint64_t d = rowoff[u + 1] - rowoff[u];
        if (d > maxdeg) maxdeg = d;
        for (uint64_t e = rowoff[u]; e < rowoff[u + 1]; e++) {
            if (cols[e] >= n) return ORC_ERANGE;
            if (e > rowoff[u] && cols[e] <= cols[e - 1]) return ORC_EUNSORTED;
        }
    }
    uint32_t *a = (uint32_t *)malloc(sizeof(uint32_t) * (maxdeg + 1));
    uint32_t *b = (uint32_t *)malloc(sizeof(uint32_t) * (maxdeg + 1));
    uint32_t *c = (uint32_t *)malloc(sizeof(uint32_t) * (maxdeg + 1));
    bitbuf bb = {0};
    int st = ORC_OK;
    if (!a || !b || !c) st = ORC_ENOMEM;
    for (uint64_t u = 0; u < n && st == ORC_OK; u++) {
        bit_offsets[u] = bb.nbits;
        st = encode_vertex(&bb, u, cols + rowoff[u], rowoff[u + 1] - rowoff[u], minLen, segLen, (int)k, 0, a, b,
                           c);
        if (bb.oom) st = ORC_ENOMEM;
    }
    free(a); free(b); free(c);
    if (st != ORC_OK) { free(bb.buf); return st; }
    bit_offsets[n] = bb.nbits;
    if (!bb.buf) bb.buf = (uint8_t *)calloc(1, 1);
    *bytes_out = bb.buf;
    *nbits_out = bb.nbits;
    return ORC_OK;
}

/* The records of vertices [u0, u1) as a standalone bit stream (R2 concatenation), for the per-vertex-parallel
 * encoder of gcgt_oracle_par.c ("per-vertex parallel with a prefix sum").  rel_offsets[i] = start
 * of u0+i relative to the chunk (u1-u0 entries).  Rows are assumed validated (orc_encode_par validates first). */
int orc_encode_range(const uint64_t *rowoff, const uint32_t *cols, uint32_t minLen, uint32_t segLen, uint32_t k,
                     uint64_t u0, uint64_t u1, uint8_t **bytes_out, uint64_t *nbits_out, uint64_t *rel_offsets) {
    uint64_t maxdeg = 0;
    for (uint64_t u = u0; u < u1; u++) if (rowoff[u + 1] - rowoff[u] > maxdeg) maxdeg = rowoff[u + 1] - rowoff[u];
    uint32_t *a = (uint32_t *)malloc(sizeof(uint32_t) * (maxdeg + 1));
    uint32_t *b = (uint32_t *)malloc(sizeof(uint32_t) * (maxdeg + 1));
    uint32_t *c = (uint32_t *)malloc(sizeof(uint32_t) * (maxdeg + 1));
    bitbuf bb = {0};
    int st = (a && b && c) ? ORC_OK : ORC_ENOMEM;
    for (uint64_t u = u0; u < u1 && st == ORC_OK; u++) {
        rel_offsets[u - u0] = bb.nbits;
        st = encode_vertex(&bb, u, cols + rowoff[u], rowoff[u + 1] - rowoff[u], minLen, segLen, (int)k, 0, a, b, c);
        if (bb.oom) st = ORC_ENOMEM;
    }
    free(a); free(b); free(c);
    if (st != ORC_OK) { free(bb.buf); return st; }
    *bytes_out = bb.buf;
    *nbits_out = bb.nbits;
    return ORC_OK;
}

/* Encodes one vertex record standalone (u, sorted list adj[0..deg-1]) for the hand-worked pins.  Returns the bit
 * length (>= 0) and writes the bits as a '0'/'1' string into out (cap chars), or a negative status.  This is the only
 * entry that accepts illustrative != 0 (Fig. 2's pre-App. C mode, gamma, unsegmented). */
int64_t orc_encode_list(uint64_t u, const uint32_t *adj, uint64_t deg, uint32_t minLen, uint32_t segLen, uint32_t k,
                        int illustrative, char *out, uint64_t cap) {
    if (minLen == 1 || k < 1 || k > 5) return ORC_EINVAL;
    for (uint64_t e = 1; e < deg; e++) if (adj[e] <= adj[e - 1]) return ORC_EUNSORTED;
    uint32_t *a = (uint32_t *)malloc(sizeof(uint32_t) * (deg + 1));
    uint32_t *b = (uint32_t *)malloc(sizeof(uint32_t) * (deg + 1));
    uint32_t *c = (uint32_t *)malloc(sizeof(uint32_t) * (deg + 1));
    bitbuf bb = {0};
    int st = (a && b && c) ? encode_vertex(&bb, u, adj, deg, minLen, segLen, (int)k, illustrative, a, b, c)
                           : ORC_ENOMEM;
    free(a); free(b); free(c);
    if (st == ORC_OK && (bb.oom || bb.nbits + 1 > cap)) st = ORC_ENOMEM;
    if (st != ORC_OK) { free(bb.buf); return st; }
    for (uint64_t i = 0; i < bb.nbits; i++) out[i] = (char)('0' + bit_at(bb.buf, i));
    out[bb.nbits] = 0;
    int64_t n = (int64_t)bb.nbits;
    free(bb.buf);
    return n;
}

void orc_free(void *p) { free(p); }

/* ------------------------------------------------------------------------------------------------------------ */
/* Decoder: inverse of R8-R18 (Alg. 1 getNextNeighbor :545-589 for field order).                                  */
/* ------------------------------------------------------------------------------------------------------------ */

/* Decodes u's record starting at bit `start`; writes the sorted neighbour list into out[0..*deg-1] (cap entries).
 * Intervals and residuals interleave in id order, so the two sequences are merged. */
int orc_decode_vertex(const uint8_t *bytes, uint64_t nbits, uint64_t start, uint64_t u, uint32_t minLen,
                      uint32_t segLen, uint32_t k, uint32_t *out, uint64_t cap, uint64_t *deg_out,
                      uint64_t *end_out) {
    uint64_t p = start, v, deg = 0, itvNum, total_itv = 0;
    int kk = (int)k;
    if (segLen == 0) { if (orc_vlc_read(kk, bytes, nbits, &p, &v) || v < 1) return ORC_EFORMAT; deg = v - 1; }
    if (orc_vlc_read(kk, bytes, nbits, &p, &v) || v < 1) return ORC_EFORMAT;
    itvNum = v - 1;
    /* Intervals first into a scratch area at the end of out, then residuals; finally merge. */
    uint64_t nout = 0;
    int64_t prev_end = 0;
    uint64_t *is = (uint64_t *)malloc(sizeof(uint64_t) * (itvNum + 1));
    uint64_t *il = (uint64_t *)malloc(sizeof(uint64_t) * (itvNum + 1));
    if (!is || !il) { free(is); free(il); return ORC_ENOMEM; }
    for (uint64_t t = 0; t < itvNum; t++) {
        uint64_t g, l;
        if (orc_vlc_read(kk, bytes, nbits, &p, &g) || orc_vlc_read(kk, bytes, nbits, &p, &l)) goto bad;
        int64_t s;
        if (t == 0) { uint64_t z = g - 1; s = (int64_t)u + ((z & 1) ? -(int64_t)(z >> 1) : (int64_t)(z >> 1)); }  /* R9 */
        else s = prev_end + (int64_t)g;                                                                    /* R10 */
        uint64_t len = l - 1 + minLen;
        is[t] = (uint64_t)s; il[t] = len;
        prev_end = s + (int64_t)len - 1;
        total_itv += len;
    }
    /* Residuals. */
    uint64_t nres_total = 0;
    uint32_t *res = NULL;
    if (segLen == 0) {
        if (deg < total_itv) goto bad;
        nres_total = deg - total_itv;
        res = (uint32_t *)malloc(sizeof(uint32_t) * (nres_total + 1));
        if (!res) goto bad;
        int64_t cur = 0;
        for (uint64_t t = 0; t < nres_total; t++) {
            if (orc_vlc_read(kk, bytes, nbits, &p, &v)) { free(res); goto bad; }
            if (t == 0) { uint64_t z = v - 1; cur = (int64_t)u + ((z & 1) ? -(int64_t)(z >> 1) : (int64_t)(z >> 1)); }  /* R11 */
            else cur += (int64_t)v;                                                                               /* R12 */
            res[t] = (uint32_t)cur;
        }
    } else {
        uint64_t segBits = 8ull * segLen, segNum;
        if (orc_vlc_read(kk, bytes, nbits, &p, &v) || v < 1) goto bad;
        segNum = v - 1;
        uint64_t base = p, cap_res = 0;
        res = NULL;
        for (uint64_t s = 0; s < segNum; s++) {                                   /* R16: segment s at base+s*segBits */
            uint64_t q = base + s * segBits, cnt;
            if (orc_vlc_read(kk, bytes, nbits, &q, &v) || v < 2) { free(res); goto bad; }
            cnt = v - 1;
            if (nres_total + cnt > cap_res) {
                cap_res = 2 * (nres_total + cnt);
                uint32_t *nr = (uint32_t *)realloc(res, sizeof(uint32_t) * cap_res);
                if (!nr) { free(res); goto bad; }
                res = nr;
            }
            int64_t cur = 0;
            for (uint64_t t = 0; t < cnt; t++) {                                  /* R17 */
                if (orc_vlc_read(kk, bytes, nbits, &q, &v)) { free(res); goto bad; }
                if (t == 0) { uint64_t z = v - 1; cur = (int64_t)u + ((z & 1) ? -(int64_t)(z >> 1) : (int64_t)(z >> 1)); }
                else cur += (int64_t)v;
                res[nres_total++] = (uint32_t)cur;
            }
            if (s + 1 == segNum) p = q;                                           /* record ends after last seg */
        }
        if (segNum == 0) p = base;
        deg = total_itv + nres_total;
    }
    if (deg > cap) { free(res); goto bad; }
    /* Merge intervals and residuals (both ascending). */
    {
        uint64_t ti = 0, off = 0, tr = 0;
        while (ti < itvNum || tr < nres_total) {
            uint64_t iv = ti < itvNum ? is[ti] + off : UINT64_MAX;
            uint64_t rv = tr < nres_total ? res[tr] : UINT64_MAX;
            if (iv < rv) { out[nout++] = (uint32_t)iv; if (++off == il[ti]) { ti++; off = 0; } }
            else { out[nout++] = (uint32_t)rv; tr++; }
        }
    }
    free(res); free(is); free(il);
    *deg_out = nout;
    if (end_out) *end_out = p;
    return ORC_OK;
bad:
    free(is); free(il);
    return ORC_EFORMAT;
}

/* Full decode into CSR.  rowoff_out: n+1 entries; cols_out: cap entries. */
int orc_decode(uint64_t n, const uint8_t *bytes, const uint64_t *bit_offsets, uint32_t minLen, uint32_t segLen,
               uint32_t k, uint64_t *rowoff_out, uint32_t *cols_out, uint64_t cap) {
    uint64_t nbits = bit_offsets[n], m = 0;
    rowoff_out[0] = 0;
    for (uint64_t u = 0; u < n; u++) {
        uint64_t d = 0, end = 0;
        int st = orc_decode_vertex(bytes, nbits, bit_offsets[u], u, minLen, segLen, k, cols_out + m, cap - m, &d, &end);
        if (st) return st;
        if (end != bit_offsets[u + 1]) return ORC_EFORMAT;            /* records are contiguous (R2) */
        m += d;
        rowoff_out[u + 1] = m;
    }
    return ORC_OK;
}

/* ------------------------------------------------------------------------------------------------------------ */
/* Alg. 4 parallelDecode, emulated step by step (Ex. 5.1 / Fig. 5 :992-1050).                 */
/* ------------------------------------------------------------------------------------------------------------ */
/* K threads start decoding (gamma, k = zeta_k) at bits 0..K-1 of the window.  vals[i], poss0[i] = decoded value and
 * bit after it (relative to the window, -1 if the codeword runs past nbits).  Then the marking rounds of lines 9-15:
 * trace_poss / trace_flags receive K entries per round r = 0..max_rounds-1 (round 0 = the initial state), with
 * -1 standing for Fig. 5's 'x' (stale / >= K).  Returns the number of rounds recorded (the initial state plus one
 * per marking round, stopping when no flagged thread has pos < K, line 12).  results[] gets the valid values in
 * order (exclusiveSum, lines 16-17) and *total their count. */
int orc_alg4_trace(int k, const uint8_t *bytes, uint64_t nbits, int K, int max_rounds, uint64_t *vals,
                   int64_t *trace_poss, int32_t *trace_flags, uint64_t *results, int *total) {
    if (K <= 0 || K > 1024) return -1;
    int64_t *poss = (int64_t *)malloc(sizeof(int64_t) * K), *np = (int64_t *)malloc(sizeof(int64_t) * K);
    int32_t *flags = (int32_t *)malloc(sizeof(int32_t) * K), *nf = (int32_t *)malloc(sizeof(int32_t) * K);
    for (int i = 0; i < K; i++) {                                          /* lines 5-8 */
        uint64_t p = (uint64_t)i, v = 0;
        if ((uint64_t)i < nbits && orc_vlc_read(k, bytes, nbits, &p, &v) == 0) { vals[i] = v; poss[i] = (int64_t)p; }
        else { vals[i] = 0; poss[i] = -1; }
        flags[i] = i == 0 ? 1 : 0;
    }
    int r = 0;
    for (;;) {
        if (r < max_rounds) {
            for (int i = 0; i < K; i++) {
                trace_poss[(int64_t)r * K + i] = poss[i];
                trace_flags[(int64_t)r * K + i] = flags[i];
            }
        }
        r++;
        int any = 0;                                                       /* line 12: syncNone(flag && pos<K) */
        for (int i = 0; i < K; i++) if (flags[i] && poss[i] >= 0 && poss[i] < K) any = 1;
        if (!any) break;
        memcpy(nf, flags, sizeof(int32_t) * K);
        for (int i = 0; i < K; i++) {                                      /* lines 13-15 */
            if (poss[i] >= 0 && poss[i] < K) {
                if (flags[i]) nf[poss[i]] = 1;
                np[i] = poss[poss[i]];
            } else {
                np[i] = -1;                                                /* 'x' propagates */
            }
        }
        memcpy(flags, nf, sizeof(int32_t) * K);
        memcpy(poss, np, sizeof(int64_t) * K);
    }
    int t = 0;                                                             /* lines 16-17 */
    for (int i = 0; i < K; i++) if (flags[i]) results[t++] = vals[i];
    *total = t;
    free(poss); free(np); free(flags); free(nf);
    return r;
}

/* ------------------------------------------------------------------------------------------------------------ */
/* Applications (§6 :1137-1286, Fig. 7).  All take a plain CSR (n, rowoff[n+1], cols[m]) of out-arcs.             */
/* ------------------------------------------------------------------------------------------------------------ */

/* BFS levels by FIFO queue (Fig. 7(b) :1143-1149).  levels[v] = hop distance from source, -1 if unreached. */
int orc_bfs(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, uint64_t source, int32_t *levels) {
    if (source >= n) return ORC_ERANGE;
    uint32_t *q = (uint32_t *)malloc(sizeof(uint32_t) * (n + 1));
    if (!q) return ORC_ENOMEM;
    for (uint64_t v = 0; v < n; v++) levels[v] = -1;
    uint64_t head = 0, tail = 0;
    levels[source] = 0; q[tail++] = (uint32_t)source;
    while (head < tail) {
        uint32_t u = q[head++];
        for (uint64_t e = rowoff[u]; e < rowoff[u + 1]; e++) {
            uint32_t v = cols[e];
            if (levels[v] < 0) { levels[v] = levels[u] + 1; q[tail++] = v; }
        }
    }
    free(q);
    return ORC_OK;
}

/* BFS that decodes the CGR on the fly, vertex by vertex (the paper's "Naive" single-thread role, :1324-1329). */
int orc_bfs_cgr(uint64_t n, const uint8_t *bytes, const uint64_t *bit_offsets, uint32_t minLen, uint32_t segLen,
                uint32_t k, uint64_t source, int32_t *levels, uint64_t *edges_out) {
    if (source >= n) return ORC_ERANGE;
    uint32_t *q = (uint32_t *)malloc(sizeof(uint32_t) * (n + 1));
    uint64_t cap = 1024;
    uint32_t *adj = (uint32_t *)malloc(sizeof(uint32_t) * cap);
    if (!q || !adj) { free(q); free(adj); return ORC_ENOMEM; }
    for (uint64_t v = 0; v < n; v++) levels[v] = -1;
    uint64_t head = 0, tail = 0, edges = 0, nbits = bit_offsets[n];
    levels[source] = 0; q[tail++] = (uint32_t)source;
    while (head < tail) {
        uint32_t u = q[head++];
        uint64_t d = 0;
        int st;
        while ((st = orc_decode_vertex(bytes, nbits, bit_offsets[u], u, minLen, segLen, k, adj, cap, &d, NULL)) ==
               ORC_EFORMAT && cap < (1ull << 34)) {
            /* the list may simply be longer than the scratch buffer: grow and retry */
            uint64_t ncap = cap * 4;
            uint32_t *na = (uint32_t *)realloc(adj, sizeof(uint32_t) * ncap);
            if (!na) break;
            adj = na; cap = ncap;
            if (cap > n + 1 && cap > 4 * (n + 1)) break;
        }
        if (st) { free(q); free(adj); return st; }
        edges += d;
        for (uint64_t e = 0; e < d; e++) {
            uint32_t v = adj[e];
            if (levels[v] < 0) { levels[v] = levels[u] + 1; q[tail++] = v; }
        }
    }
    free(q); free(adj);
    if (edges_out) *edges_out = edges;
    return ORC_OK;
}

/* Weakly connected components by sequential union-find (disjoint-set forests [19], :1256-1271); every arc joins
 * both endpoints; labels[v] = minimum vertex id of v's component (north_star). */
static uint64_t uf_find(uint32_t *parent, uint64_t x) {
    while (parent[x] != x) x = parent[x];
    return x;
}

int orc_cc(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, uint32_t *labels) {
    uint32_t *parent = labels;                      /* union by min root: the root is always the set's minimum */
    for (uint64_t v = 0; v < n; v++) parent[v] = (uint32_t)v;
    for (uint64_t u = 0; u < n; u++) {
        for (uint64_t e = rowoff[u]; e < rowoff[u + 1]; e++) {
            uint64_t ru = uf_find(parent, u), rv = uf_find(parent, cols[e]);
            if (ru < rv) parent[rv] = (uint32_t)ru;
            else if (rv < ru) parent[ru] = (uint32_t)rv;
        }
        /* path compression of u's chain keeps find() cheap; it never changes any root */
        uint64_t r = uf_find(parent, u), x = u;
        while (parent[x] != x) { uint64_t nx = parent[x]; parent[x] = (uint32_t)r; x = nx; }
    }
    for (uint64_t v = 0; v < n; v++) labels[v] = (uint32_t)uf_find(parent, v);
    return ORC_OK;
}

/* Betweenness centrality, textbook Brandes [9] (§6 :1272-1284, Fig. 7(d) :1243-1244).  For each source s
 * (duplicates counted): BFS over out-arcs gives d and sigma; then, over vertices in reverse BFS order,
 *   delta(v) = sum_{w in out(v), d(w) = d(v)+1} sigma(v)/sigma(w) * (1 + delta(w))   (Fig. 7(d)'s formula)
 * and bc[v] += delta(v) for v != s.  Unnormalised, not halved; fp64. */
int orc_bc(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, const uint32_t *sources, uint64_t nsrc,
           double *bc) {
    int32_t *d = (int32_t *)malloc(sizeof(int32_t) * n);
    double *sigma = (double *)malloc(sizeof(double) * n), *delta = (double *)malloc(sizeof(double) * n);
    uint32_t *S = (uint32_t *)malloc(sizeof(uint32_t) * (n + 1));
    if (!d || !sigma || !delta || !S) { free(d); free(sigma); free(delta); free(S); return ORC_ENOMEM; }
    for (uint64_t v = 0; v < n; v++) bc[v] = 0.0;
    for (uint64_t si = 0; si < nsrc; si++) {
        uint64_t s = sources[si];
        if (s >= n) { free(d); free(sigma); free(delta); free(S); return ORC_ERANGE; }
        for (uint64_t v = 0; v < n; v++) { d[v] = -1; sigma[v] = 0.0; delta[v] = 0.0; }
        uint64_t head = 0, tail = 0;
        d[s] = 0; sigma[s] = 1.0; S[tail++] = (uint32_t)s;
        while (head < tail) {                                   /* forward pass: distance and sigma */
            uint32_t v = S[head++];
            for (uint64_t e = rowoff[v]; e < rowoff[v + 1]; e++) {
                uint32_t w = cols[e];
                if (d[w] < 0) { d[w] = d[v] + 1; S[tail++] = w; }
                if (d[w] == d[v] + 1) sigma[w] += sigma[v];
            }
        }
        for (uint64_t i = tail; i-- > 0;) {                     /* backward pass, descending distance */
            uint32_t v = S[i];
            double acc = 0.0;
            for (uint64_t e = rowoff[v]; e < rowoff[v + 1]; e++) {
                uint32_t w = cols[e];
                if (d[w] == d[v] + 1) acc += sigma[v] / sigma[w] * (1.0 + delta[w]);
            }
            delta[v] = acc;
            if (v != s) bc[v] += acc;
        }
    }
    free(d); free(sigma); free(delta); free(S);
    return ORC_OK;
}

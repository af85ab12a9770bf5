/*
 * gcgt_oracle_par.c — the oracle's multi-threaded BFS (OpenMP), for host-side timing and full-size parity.
 *
 * TEST INFRASTRUCTURE ONLY (same rules as gcgt_oracle.c): only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load it; it shares nothing with the product path.
 *
 * SURVEY §8(c).2 "Host parallelism for timing": a level-synchronous variant of the FIFO BFS over the same decoder.
 * BFS levels are unique (the hop distance), so the result equals orc_bfs / orc_bfs_cgr exactly; this is the role
 * Ligra / Ligra+ play in the paper's Fig. 8 (36 host cores).
 * Level d: every frontier vertex u is expanded (its record decoded with orc_decode_vertex, or its CSR row read);
 * each neighbour v with level -1 is claimed by one compare-and-swap -1 -> d+1, and the winner appends v to its
 * thread's next-frontier list; the lists are concatenated into the next frontier.
 * Pin: tests/test_oracle_algos.py (equal to orc_bfs on random graphs, on every recipe, for 1..8 threads).
 */
#include <omp.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

enum { PAR_OK = 0, PAR_ERANGE = -3, PAR_ENOMEM = -5, PAR_EFORMAT = -8 };

int orc_decode_vertex(const uint8_t *bytes, uint64_t nbits, uint64_t start, uint64_t u, uint32_t minLen,
                      uint32_t segLen, uint32_t k, uint32_t *out, uint64_t cap, uint64_t *deg_out,
                      uint64_t *end_out);

typedef struct { uint32_t *v; uint64_t n, cap; } vec32;

static int vpush(vec32 *a, uint32_t x) {
    if (a->n == a->cap) {
        uint64_t nc = a->cap ? 2 * a->cap : 4096;
        uint32_t *nv = (uint32_t *)realloc(a->v, sizeof(uint32_t) * nc);
        if (!nv) return -1;
        a->v = nv; a->cap = nc;
    }
    a->v[a->n++] = x;
    return 0;
}

static int claim(int32_t *levels, uint32_t v, int32_t d1) {
    int32_t expect = -1;
    if (__atomic_load_n(&levels[v], __ATOMIC_RELAXED) != -1) return 0;
    return __atomic_compare_exchange_n(&levels[v], &expect, d1, 0, __ATOMIC_RELAXED, __ATOMIC_RELAXED);
}

static void seterr(int *err, int st) { __atomic_store_n(err, st, __ATOMIC_RELAXED); }

/* Shared level loop.  csr != 0: rows from (rowoff, cols); else records decoded from the CGR. */
static int bfs_levels(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, const uint8_t *bytes,
                      const uint64_t *offs, uint32_t minLen, uint32_t segLen, uint32_t k, uint64_t source,
                      int32_t *levels, uint64_t *edges_out, int nthreads, uint64_t max_edges) {
    if (source >= n) return PAR_ERANGE;
    if (nthreads > 0) omp_set_num_threads(nthreads);
    const int T = nthreads > 0 ? nthreads : omp_get_max_threads();
#pragma omp parallel for schedule(static)
    for (int64_t v = 0; v < (int64_t)n; v++) levels[v] = -1;
    uint32_t *front = (uint32_t *)malloc(sizeof(uint32_t) * (n + 1));
    vec32 *next = (vec32 *)calloc((size_t)T, sizeof(vec32));
    if (!front || !next) { free(front); free(next); return PAR_ENOMEM; }
    uint64_t nf = 1, edges = 0;
    int err = PAR_OK;
    front[0] = (uint32_t)source;
    levels[source] = 0;
    for (int32_t d = 0; nf && !err && edges < max_edges; d++) {
#pragma omp parallel num_threads(T) reduction(+ : edges)
        {
            const int t = omp_get_thread_num();
            vec32 *mine = &next[t];
            mine->n = 0;
            uint64_t cap = 1024;
            uint32_t *adj = bytes ? (uint32_t *)malloc(sizeof(uint32_t) * cap) : NULL;
#pragma omp for schedule(dynamic, 64)
            for (int64_t i = 0; i < (int64_t)nf; i++) {
                const uint32_t u = front[i];
                if (!bytes) {
                    edges += rowoff[u + 1] - rowoff[u];
                    for (uint64_t e = rowoff[u]; e < rowoff[u + 1]; e++)
                        if (claim(levels, cols[e], d + 1) && vpush(mine, cols[e])) seterr(&err, PAR_ENOMEM);
                    continue;
                }
                uint64_t deg = 0;
                int st;
                while (adj && (st = orc_decode_vertex(bytes, offs[n], offs[u], u, minLen, segLen, k, adj, cap,
                                                      &deg, NULL)) == PAR_EFORMAT && cap <= 4 * (n + 1)) {
                    cap *= 4;  /* the list may be longer than the scratch buffer: grow and retry */
                    uint32_t *na = (uint32_t *)realloc(adj, sizeof(uint32_t) * cap);
                    if (!na) { free(adj); adj = NULL; }
                    else adj = na;
                }
                if (!adj) { seterr(&err, PAR_ENOMEM); continue; }
                if (st) { seterr(&err, st); continue; }
                edges += deg;
                for (uint64_t e = 0; e < deg; e++)
                    if (claim(levels, adj[e], d + 1) && vpush(mine, adj[e])) seterr(&err, PAR_ENOMEM);
            }
            free(adj);
        }
        uint64_t tot = 0;
        for (int t = 0; t < T; t++) {
            memcpy(front + tot, next[t].v, sizeof(uint32_t) * next[t].n);
            tot += next[t].n;
        }
        nf = tot;
    }
    for (int t = 0; t < T; t++) free(next[t].v);
    free(next);
    free(front);
    if (edges_out) *edges_out = edges;
    return err;
}

/* BFS over the oracle's own CGR (decoded vertex by vertex), nthreads threads (0 = all cores). */
int orc_bfs_cgr_par(uint64_t n, const uint8_t *bytes, const uint64_t *bit_offsets, uint32_t minLen, uint32_t segLen,
                    uint32_t k, uint64_t source, int32_t *levels, uint64_t *edges_out, int nthreads) {
    return bfs_levels(n, NULL, NULL, bytes, bit_offsets, minLen, segLen, k, source, levels, edges_out, nthreads,
                      UINT64_MAX);
}

/* Bounded sample of the same BFS for timing: whole levels are expanded until at least max_edges arcs have been
 * decoded (*edges_out = arcs decoded; the levels of later vertices are left incomplete). */
int orc_bfs_cgr_sample(uint64_t n, const uint8_t *bytes, const uint64_t *bit_offsets, uint32_t minLen,
                       uint32_t segLen, uint32_t k, uint64_t source, int32_t *levels, uint64_t *edges_out,
                       int nthreads, uint64_t max_edges) {
    return bfs_levels(n, NULL, NULL, bytes, bit_offsets, minLen, segLen, k, source, levels, edges_out, nthreads,
                      max_edges);
}

/* The same level loop over a plain CSR (full-size parity of the largest configs, where decoding would only repeat
 * what the round-trip pins already establish). */
int orc_bfs_par(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, uint64_t source, int32_t *levels,
                int nthreads) {
    return bfs_levels(n, rowoff, cols, NULL, NULL, 0, 0, 0, source, levels, NULL, nthreads, UINT64_MAX);
}

int orc_max_threads(void) { return omp_get_max_threads(); }

/* ---- encoder, per-vertex parallel with a prefix sum -------------------------------------------
 * The vertex range is cut into chunks; each chunk's records are encoded by orc_encode_range (the same per-vertex
 * encode_vertex as orc_encode), then the chunks are concatenated at the prefix sum of their bit lengths (R2).
 * Pin: byte-identical to orc_encode (tests/test_oracle_codec.py). */
int orc_encode_range(const uint64_t *rowoff, const uint32_t *cols, uint32_t minLen, uint32_t segLen, uint32_t k,
                     uint64_t u0, uint64_t u1, uint8_t **bytes_out, uint64_t *nbits_out, uint64_t *rel_offsets);

int orc_encode_par(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, uint32_t minLen, uint32_t segLen,
                   uint32_t k, uint8_t **bytes_out, uint64_t *nbits_out, uint64_t *bit_offsets, int nthreads) {
    if (minLen == 1 || k < 1 || k > 5) return -1;
    if (nthreads > 0) omp_set_num_threads(nthreads);
    int bad = 0;
#pragma omp parallel for schedule(dynamic, 4096) reduction(| : bad)
    for (int64_t u = 0; u < (int64_t)n; u++) {                       /* R6: validate every row */
        if (rowoff[u + 1] < rowoff[u]) { bad |= 1; continue; }
        for (uint64_t e = rowoff[u]; e < rowoff[u + 1]; e++) {
            if (cols[e] >= n) bad |= 2;
            else if (e > rowoff[u] && cols[e] <= cols[e - 1]) bad |= 4;
        }
    }
    if (bad & 1) return -1;
    if (bad & 2) return PAR_ERANGE;
    if (bad & 4) return -2;
    const uint64_t chunk = 1 << 16, nch = (n + chunk - 1) / chunk;
    uint8_t **cb = (uint8_t **)calloc(nch + 1, sizeof(uint8_t *));
    uint64_t *cn = (uint64_t *)calloc(nch + 1, sizeof(uint64_t));
    if (!cb || !cn) { free(cb); free(cn); return PAR_ENOMEM; }
    int err = PAR_OK;
#pragma omp parallel for schedule(dynamic, 1)
    for (int64_t c = 0; c < (int64_t)nch; c++) {
        const uint64_t u0 = (uint64_t)c * chunk, u1 = u0 + chunk < n ? u0 + chunk : n;
        const int st = orc_encode_range(rowoff, cols, minLen, segLen, k, u0, u1, &cb[c], &cn[c], bit_offsets + u0);
        if (st) seterr(&err, st);
    }
    uint64_t total = 0;
    for (uint64_t c = 0; c < nch; c++) { const uint64_t l = cn[c]; cn[c] = total; total += l; }
    cn[nch] = total;
    uint8_t *out = err ? NULL : (uint8_t *)calloc(total / 8 + 2, 1);
    if (!out && !err) err = PAR_ENOMEM;
    if (!err) {
#pragma omp parallel for schedule(dynamic, 1)
        for (int64_t c = 0; c < (int64_t)nch; c++) {
            const uint64_t u0 = (uint64_t)c * chunk, u1 = u0 + chunk < n ? u0 + chunk : n;
            const uint64_t base = cn[c], len = cn[c + 1] - cn[c], sh = base & 7;
            for (uint64_t u = u0; u < u1; u++) bit_offsets[u] += base;
            /* MSB-first (R1): source byte j lands in destination bytes base/8 + j (>> sh) and + j + 1 (<< 8-sh);
             * chunk boundary bytes are shared with the neighbours, so every store is an atomic OR */
            for (uint64_t j = 0; j < (len + 7) / 8; j++) {
                uint8_t x = cb[c][j];
                if (j == len / 8) x &= (uint8_t)(0xFF00u >> (len & 7));   /* only the chunk's own bits */
                if (!x) continue;
                __atomic_fetch_or(&out[base / 8 + j], (uint8_t)(x >> sh), __ATOMIC_RELAXED);
                if (sh) __atomic_fetch_or(&out[base / 8 + j + 1], (uint8_t)(x << (8 - sh)), __ATOMIC_RELAXED);
            }
        }
    }
    for (uint64_t c = 0; c < nch; c++) free(cb[c]);
    free(cb);
    free(cn);
    if (err) { free(out); return err; }
    bit_offsets[n] = total;
    *bytes_out = out;
    *nbits_out = total;
    return PAR_OK;
}

/* ---- Brandes BC, parallel over sources -------------------------------------------------------
 * Each source's dependencies delta_s are computed by the same textbook Brandes as orc_bc (one source at a time per
 * thread, orc_bc with nsrc = 1 into a private vector); the per-source vectors are then summed in source order, so
 * the result is bit-identical to orc_bc.  Pin: tests/test_oracle_algos.py. */
int orc_bc(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, const uint32_t *sources, uint64_t nsrc,
           double *bc);

int orc_bc_par(uint64_t n, const uint64_t *rowoff, const uint32_t *cols, const uint32_t *sources, uint64_t nsrc,
               double *bc, int nthreads) {
    if (nthreads > 0) omp_set_num_threads(nthreads);
    for (uint64_t v = 0; v < n; v++) bc[v] = 0.0;
    const int T = nthreads > 0 ? nthreads : omp_get_max_threads();
    const uint64_t B = (uint64_t)T;  /* sources per round: one private vector per thread */
    double *part = (double *)malloc(sizeof(double) * (n ? n : 1) * B);
    if (!part) return PAR_ENOMEM;
    int err = PAR_OK;
    for (uint64_t s0 = 0; s0 < nsrc && !err; s0 += B) {
        const uint64_t cnt = nsrc - s0 < B ? nsrc - s0 : B;
#pragma omp parallel for schedule(dynamic, 1) num_threads(T)
        for (int64_t i = 0; i < (int64_t)cnt; i++) {
            const int st = orc_bc(n, rowoff, cols, sources + s0 + i, 1, part + (uint64_t)i * n);
            if (st) seterr(&err, st);
        }
        for (uint64_t i = 0; i < cnt; i++) {                            /* source order */
            const double *p = part + i * n;
#pragma omp parallel for schedule(static)
            for (int64_t v = 0; v < (int64_t)n; v++) bc[v] += p[v];
        }
    }
    free(part);
    return err;
}

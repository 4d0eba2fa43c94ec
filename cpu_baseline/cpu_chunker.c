/*
 * cpu_chunker.c — multithreaded CPU rolling Rabin chunker: the CPU baseline that north_star
 * asks to time beside the GPU (not the oracle, not the product).
 *
 * The paper's host-only design (§5.1): "(1) divide the input data equally
 * in fixed-size regions among N threads; (2) invoke the Rabin fingerprint-based chunking
 * algorithm in parallel on N different regions; (3) synchronize neighboring threads in the end
 * to merge the resulting chunk boundaries".  Each region re-reads the w-1 bytes before it (the
 * window overlap, L282-L287), rolls f <- ((f << 8) mod x^k) ^ b ^ T[top byte] ^ U[out byte],
 * and keeps its candidates; the lists are concatenated in region order; the min/max rule runs
 * once over the result.  Tables are built here with their own GF(2) code.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#include <pthread.h>

typedef struct {
    const uint8_t *d; uint64_t n, lo, hi;       /* window ends [lo, hi) */
    uint32_t w; int k; uint64_t kmask, dmask, r;
    const uint64_t *T, *U;
    uint64_t *list; uint64_t cnt, cap;
} job_t;

static int deg(uint64_t p) { int d = -1; for (int t = 0; t < 64; ++t) if ((p >> t) & 1) d = t; return d; }

static void tables(uint64_t P, int k, uint32_t w, uint64_t *T, uint64_t *U) {
    /* x^e mod P by repeated multiplication by x */
    uint64_t xk[8], xw[8], v = 1;
    uint64_t e = 0, target = (uint64_t)k, tw = 8ull * w;
    uint64_t hi = (uint64_t)1 << k;
    for (; e < target; ++e) { v <<= 1; if (v & hi) v ^= P; }
    for (int j = 0; j < 8; ++j) { xk[j] = v; v <<= 1; if (v & hi) v ^= P; ++e; }
    v = 1;
    for (e = 0; e < tw; ++e) { v <<= 1; if (v & hi) v ^= P; }
    for (int j = 0; j < 8; ++j) { xw[j] = v; v <<= 1; if (v & hi) v ^= P; }
    for (int t = 0; t < 256; ++t) {
        uint64_t a = 0, b = 0;
        for (int j = 0; j < 8; ++j) if ((t >> j) & 1) { a ^= xk[j]; b ^= xw[j]; }
        T[t] = a; U[t] = b;
    }
}

static void *work(void *arg) {
    job_t *J = (job_t *)arg;
    const uint8_t *d = J->d;
    uint64_t p = J->lo >= J->w - 1 ? J->lo - (J->w - 1) : 0;
    uint64_t f = 0;
    const int sh = J->k - 8;
    for (uint64_t i = p; i < J->hi; ++i) {
        f = ((f << 8) & J->kmask) ^ d[i] ^ J->T[(f >> sh) & 0xff];
        if (i >= p + J->w) f ^= J->U[d[i - J->w]];
        if (i >= J->lo && (f & J->dmask) == J->r && i + 1 < J->n && i + 1 >= J->w) {
            if (J->cnt == J->cap) {
                J->cap = J->cap ? 2 * J->cap : 4096;
                J->list = (uint64_t *)realloc(J->list, J->cap * sizeof(uint64_t));
            }
            J->list[J->cnt++] = i + 1;
        }
    }
    return NULL;
}

/* Returns the number of cuts (writes min(count, cap)); threads >= 1. */
int64_t cpu_chunk(const uint8_t *d, uint64_t n, uint64_t poly, uint32_t w, uint64_t D, uint64_t r,
                  uint64_t mn, uint64_t mx, int threads, uint64_t *out, uint64_t cap) {
    uint64_t T[256], U[256];
    int k = deg(poly);
    tables(poly, k, w, T, U);
    if (threads < 1) threads = 1;
    job_t *J = (job_t *)calloc(threads, sizeof(job_t));
    pthread_t *th = (pthread_t *)calloc(threads, sizeof(pthread_t));
    for (int t = 0; t < threads; ++t) {
        J[t] = (job_t){d, n, n * t / threads, n * (t + 1) / threads, w, k,
                       (k == 64) ? ~0ull : ((1ull << k) - 1), D - 1, r, T, U, NULL, 0, 0};
        pthread_create(&th[t], NULL, work, &J[t]);
    }
    uint64_t s = 0; int64_t cnt = 0;
#define EMIT(v) do { if ((uint64_t)cnt < cap) out[cnt] = (v); ++cnt; } while (0)
    for (int t = 0; t < threads; ++t) {          /* merge in region order, then the size rule */
        pthread_join(th[t], NULL);
        for (uint64_t j = 0; j < J[t].cnt; ++j) {
            uint64_t c = J[t].list[j];
            if (!mn && !mx) { EMIT(c); continue; }
            if (mx) while (c - s > mx) { s += mx; EMIT(s); }
            if (c - s >= mn) { EMIT(c); s = c; }
        }
        free(J[t].list);
    }
    if (mx) while (n - s > mx) { s += mx; if (s < n) EMIT(s); }
#undef EMIT
    free(J); free(th);
    return cnt;
}

/*
 * splitmix_fill.c — multithreaded host filler for the counter-mode SplitMix64 input stream.
 *
 * Input generation only (synthgen/ holds no chunking arithmetic): byte j of stream `seed` is
 * byte j%8 (little-endian) of word j/8, word k = mix(seed + (k+1)*0x9E3779B97F4A7C15), the same
 * definition as synthgen.splitmix_words (numpy, the reference form) and the device's own
 * k_synth_fill.  tests/test_synthgen.py checks this filler against the numpy form.  It exists
 * because the numpy form runs at ~0.2 GB/s and the full-size configs are 16-64 GiB.
 */
#include <pthread.h>
#include <stdint.h>
#include <string.h>

static inline uint64_t sm_word(uint64_t seed, uint64_t k)
{
    uint64_t z = seed + (k + 1ull) * 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

/* bytes [off, off + len) of the stream into dst */
static void fill_range(uint8_t *dst, uint64_t len, uint64_t seed, uint64_t off)
{
    uint64_t j = 0;
    while (j < len && ((off + j) & 7u)) {                /* head up to a word boundary */
        const uint64_t p = off + j;
        dst[j++] = (uint8_t)(sm_word(seed, p >> 3) >> (8 * (p & 7u)));
    }
    for (; j + 8 <= len; j += 8) {
        const uint64_t w = sm_word(seed, (off + j) >> 3);
        uint8_t b[8];
        for (int q = 0; q < 8; ++q) b[q] = (uint8_t)(w >> (8 * q));
        memcpy(dst + j, b, 8);
    }
    for (; j < len; ++j) {
        const uint64_t p = off + j;
        dst[j] = (uint8_t)(sm_word(seed, p >> 3) >> (8 * (p & 7u)));
    }
}

typedef struct { uint8_t *dst; uint64_t len, seed, off; } job_t;

static void *worker(void *a)
{
    job_t *J = (job_t *)a;
    fill_range(J->dst, J->len, J->seed, J->off);
    return 0;
}

int sg_fill(uint8_t *dst, uint64_t len, uint64_t seed, uint64_t off, int threads)
{
    if (threads < 1) threads = 1;
    if (threads > 256) threads = 256;
    if (len < (1u << 20)) threads = 1;
    pthread_t th[256];
    int live[256];
    job_t jobs[256];
    const uint64_t per = ((len + (uint64_t)threads - 1u) / (uint64_t)threads + 7u) & ~7ull;
    int n = 0;
    for (uint64_t a = 0; a < len && n < threads; a += per, ++n) {
        const uint64_t b = a + per < len ? a + per : len;
        jobs[n].dst = dst + a; jobs[n].len = b - a; jobs[n].seed = seed; jobs[n].off = off + a;
        live[n] = pthread_create(&th[n], 0, worker, &jobs[n]) == 0;
        if (!live[n]) worker(&jobs[n]);
    }
    for (int t = 0; t < n; ++t)
        if (live[t]) pthread_join(th[t], 0);
    return 0;
}

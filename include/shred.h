/*
 * shred.h — C ABI of the B200-native content-defined chunker (Shredder's hot path).
 *
 * What it computes (PAPER.md, Bhatotia/Rodrigues/Verma, FAST'12):
 *   * L245-L258 (§2.1, Eq. (1)): a Rabin fingerprint over sliding windows of w contiguous
 *     bytes — the window, read as a polynomial over GF(2), reduced modulo an irreducible
 *     polynomial div(x) of degree k ("the remainder r(x) obtained by division of f(x)").
 *   * L444-L454 (§3.1): w = 48 bytes; a cut where the low-order 13 bits of the fingerprint
 *     equal a pre-defined marker; slide one byte forward and repeat.
 *   * L259-L269 (§2.1): min/max chunk sizes; min = 0, max = inf by default.
 *   * L416-L434 (§3.1): boundaries are handed to the application ("upcall") — here: written
 *     as ascending absolute u64 offsets into a caller buffer, on a CUDA stream.
 * Readings where the paper is silent (polynomial, marker value, bit order, cut position,
 * stream start/end, min/max off-by-ones) are DESIGN.md "Readings" Q1..Q17.
 *
 * Cut offset convention: a window ending at byte i (bytes i-w+1..i) that matches yields the
 * cut c = i+1 (exclusive end of the chunk).  Only full windows are tested (c >= w); c = N
 * (the stream end) is never emitted.  Forced max-size cuts may be < w.
 *
 * Conventions for every call:
 *   Ownership   The caller owns every pointer it passes (inputs, d_out, n_out); they must stay
 *               valid and unmodified until the work enqueued on `stream` completes.  The
 *               library owns the ctx, its device tables, scratch, ring slots, copy stream and
 *               events.  Fed bytes that must be carried (the last w-1) are copied into
 *               library memory, so a fed buffer may be reused once the call's work completes.
 *   Memory      d_* = device memory (cudaMalloc / torch CUDA tensor).  n_out = device memory or
 *               mapped page-locked host memory (cudaHostAlloc; written by a kernel).
 *   Async       Calls enqueue on `stream` and return; nothing is synchronised unless stated.
 *               Exception: a call that needs more scratch than any earlier call of the ctx
 *               grows it synchronously (cudaDeviceSynchronize before freeing the old buffer).
 *   Streams     A ctx is bound to one device and is not re-entrant (one caller thread at a
 *               time).  Its calls share the ctx's scratch, state and ring, so they run in call
 *               order: a call on a stream other than the previous call's first makes its stream
 *               wait for the work enqueued on that stream (an event; no host synchronisation).  Under
 *               CUDA-graph capture no event is recorded or waited on: capture a ctx's calls on
 *               the stream its preceding work used (or synchronise before capturing).  The
 *               previous call's stream must still exist when a call switches streams (the end
 *               of its work is recorded on it then).
 *   Errors      Negative return codes are synchronous problems (parameters, enqueue,
 *               allocation).  Output-capacity overflow is in-band: *n_out receives the TRUE
 *               count n and min(n, cap) offsets are written (snprintf convention).  In the
 *               streaming calls an overflow loses emitted offsets, so the ctx turns sticky
 *               SHRED_ECAPACITY (checked at the next call, which is refused).
 */
#ifndef SHRED_H
#define SHRED_H

#include <stdint.h>
#include <stddef.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct CUstream_st *shred_stream_t;   /* == cudaStream_t; NULL = legacy default stream */

typedef struct shred_params {
    uint64_t poly;      /* div(x) over GF(2): bit t = coefficient of x^t; irreducible,
                           8 <= deg <= 63.  Default 0xbfe6b8a5bf378d83 (deg 63, reading Q1).  */
    uint32_t window;    /* w bytes, 1 <= w <= 4096.  Default 48 (L444-L446).                   */
    uint32_t marker;    /* SHRED_MARKER_EQ (0, default): a cut candidate where fp mod D == r
                           (L447-L451); SHRED_MARKER_LE (1): where fp mod D <= r, the "value mod
                           p is lower or equal to a constant" marker set of L249-L251.          */
    uint64_t divisor;   /* D, 2 <= D <= 2^deg.  Default 8192 ("13 bits", L447).  Any other D is
                           the integer remainder of the fingerprint's value (reading Q8).  Fast
                           paths: D = 2^m <= 2^32 (either marker), or D = d 2^s with s < 32 and
                           the '==' marker (divisibility test); every other D by the remainder
                           itself (a multiply-high quotient).                                   */
    uint64_t magic;     /* r < D.  Default 0x78 (reading Q6).                                  */
    uint64_t min_size;  /* 0 = off (paper default)                                  */
    uint64_t max_size;  /* 0 = off (= inf).  Else max_size >= max(min_size, 1)                 */
} shred_params;

typedef struct shred_ctx shred_ctx;   /* opaque; bound to one CUDA device */

enum {
    SHRED_OK        =  0,
    SHRED_EINVAL    = -1,   /* bad parameter / pointer kind / length                          */
    SHRED_ENOMEM    = -2,   /* device or host allocation failed                              */
    SHRED_ECUDA     = -3,   /* a CUDA call failed at enqueue (see shred_last_error)          */
    SHRED_ESTATE    = -4,   /* misuse of the streaming state                                 */
    SHRED_ECAPACITY = -5    /* sticky: a streaming call overflowed its output buffer         */
};

enum { SHRED_MARKER_EQ = 0, SHRED_MARKER_LE = 1 };

/* Kernel paths the ctx selected for its parameters (shred_path). */
enum {
    SHRED_PATH_K63     = 1, /* deg(P) in 33..63 (the paper's reading: 63), 1 <= w <= 4096 (w > 64:
                               the bytes leaving the window from a second TMA tile), any valid D
                               and marker set (marker kinds below): u64 state, TMA-staged, smem
                               LDS.64 tables                                                    */
    SHRED_PATH_K32     = 2, /* deg(P) in 8..32, same w / D / marker conditions: u32 state, LDS.32 */
    SHRED_PATH_GENERIC = 3  /* any other valid parameters: byte-at-a-time (the hot paths also use
                               the byte loop for inputs below 4 KiB and for their edge segments) */
};

/* Fill *p with the paper defaults (readings Q1, Q5, Q6, Q15): P = 0xbfe6b8a5bf378d83, w = 48,
   D = 8192, r = 0x78, min = 0, max = 0 (off). */
void        shred_default_params(shred_params *p);

/* Validate *p (degree, irreducibility of P by Ben-Or's test, 2 <= D <= 2^deg, r < D, marker,
   min/max), build the push/pop tables (PAPER.md: "shifting a byte forward") on the
   host, upload them to `device` and create the ctx.  Synchronous.  *out = NULL on error. */
int         shred_init(const shred_params *p, int device, shred_ctx **out);

/* Synchronise the ctx's own streams and free everything it owns.  NULL is a no-op. */
void        shred_destroy(shred_ctx *ctx);

const char *shred_strerror(int code);
const char *shred_last_error(const shred_ctx *ctx);   /* detail incl. the CUDA error string  */
int         shred_path(const shred_ctx *ctx);         /* SHRED_PATH_* chosen at init          */
/* The hot kernel's state mode (diagnostics): 1 K63 (u64 state, deg 41..63), 5 K40 (deg 33..40),
   2 K32 (u32 state, T by table), 4 K32B (u32, whole-byte top byte: deg 8/16/24/32), 6 K32T (u32,
   T as one integer product: P = x^k + Q with Q's terms >= 8 apart and below k - 7, e.g. the
   trinomial x^31 + x^13 + 1; '==' and '<=' with D = 2^m), 7 K63T (the u64-state analogue for
   deg 41..63 with Q's terms below 25, e.g. x^63 + x^11 + 1), 3 generic. */
int         shred_kernel_mode(const shred_ctx *ctx);
int         shred_get_params(const shred_ctx *ctx, shred_params *out);

/* An output capacity that can never overflow for `len` input bytes:
   len-1 if min = 0 (a candidate can occur at every position), else floor((len-1)/min) + 1. */
uint64_t    shred_max_cuts(const shred_ctx *ctx, uint64_t len);

/* One-shot, device-resident chunking of d_in[0..len) as a whole stream.
   Writes the ascending final cuts (candidates, then the size rule if min > 0 or max > 0) to
   d_out[0 .. min(n, cap)) and n to *n_out.  d_in may have any alignment.  len = 0 is valid
   (n = 0).  Enqueues on `stream`, returns after enqueue (device scratch may be grown — a
   synchronous cudaMalloc — the first time a larger input is seen). */
int shred_chunk(shred_ctx *ctx, const uint8_t *d_in, uint64_t len,
                uint64_t *d_out, uint64_t cap, uint64_t *n_out, shred_stream_t stream);

/* Shard primitive for byte-range sharding (multi-GPU: "a small overlap of
   the size of the sliding window (w bytes) near partition boundaries").
   d_in points at stream position `start - halo`; the shard's own bytes are
   d_in[halo .. halo+len) = stream positions [start, start+len).  halo must equal
   min(w-1, start).  Tests every window ending at i in [start, start+len) with i >= w-1 and
   writes the cut CANDIDATES c = i+1 with c < total_len (absolute offsets, ascending) — no size
   rule — to d_out[0 .. min(n, cap)), n to *n_out. */
int shred_candidates_range(shred_ctx *ctx, const uint8_t *d_in, uint64_t halo, uint64_t start,
                           uint64_t len, uint64_t total_len,
                           uint64_t *d_out, uint64_t cap, uint64_t *n_out, shred_stream_t stream);

/* The size rule (readings Q12-Q15) over n_cand ascending candidates of a
   stream of total_len bytes (e.g. the concatenated per-shard candidate lists).  Uses the
   ctx's min/max; with both off it copies.  Writes cuts to d_out (cap, n_out as above).
   d_cand and d_out must not overlap. */
int shred_size_bound(shred_ctx *ctx, const uint64_t *d_cand, uint64_t n_cand, uint64_t total_len,
                     uint64_t *d_out, uint64_t cap, uint64_t *n_out, shred_stream_t stream);

/* The size rule from an explicit entry state over one range of the stream ending at `end`
   (the per-shard step of the distributed size rule): state_in = {s, held}
   (s = last cut; held = 1 if a cut at s is not yet emitted; {0, 0} at the stream start).
   fin = 1 if `end` is the stream end, else a candidate accepted exactly at `end` is held.
   Cuts go to d_out (cap, n_out as usual); d_state_out (device, 2 x u64) gets the exit
   {s, held}.  Chaining ranges through their states equals one run over the whole list. */
int shred_size_bound_state(shred_ctx *ctx, const uint64_t *d_cand, uint64_t n_cand, uint64_t end,
                           int fin, const uint64_t state_in[2], uint64_t *d_out, uint64_t cap,
                           uint64_t *n_out, uint64_t *d_state_out, shred_stream_t stream);

/* The same with everything the host does not need to know kept in device memory, so rounds of
   the distributed size rule chain on the stream without a host synchronisation: the candidate
   count is read from d_n_cand (device u64; at most n_cand_max, which sizes the launch), the
   entry state from d_state_in (device, 2 x u64 {s, held}).  Otherwise as above.  d_state_in and
   d_state_out may be the same array. */
int shred_size_bound_state_dev(shred_ctx *ctx, const uint64_t *d_cand, const uint64_t *d_n_cand,
                               uint64_t n_cand_max, uint64_t end, int fin, const uint64_t *d_state_in,
                               uint64_t *d_out, uint64_t cap, uint64_t *n_out, uint64_t *d_state_out,
                               shred_stream_t stream);

/* Streaming with carried window and size-rule state (§4.1-§4.2: pinned
   buffers, async transfers, multi-buffering).  `in` is device memory or page-locked host
   memory (pageable host memory -> SHRED_EINVAL).  Host input is copied by the ctx's own copy
   stream into a ring of device slots (double/triple buffering) while the previous slot is
   chunked on `stream`.  Offsets are absolute stream positions.  Only final cuts are emitted:
   a cut at exactly the current stream end is held until the next feed (emitted) or the flush
   (dropped: c = N is never a cut).  len may be 0. */
int shred_feed (shred_ctx *ctx, const void *in, uint64_t len,
                uint64_t *d_out, uint64_t cap, uint64_t *n_out, shred_stream_t stream);
/* End the stream: emits the remaining forced max-size cuts and resets the stream state. */
int shred_flush(shred_ctx *ctx, uint64_t *d_out, uint64_t cap, uint64_t *n_out,
                shred_stream_t stream);
/* Discard the stream state (synchronises the ctx's streams; clears a sticky error). */
int shred_reset(shred_ctx *ctx);
/* Ring configuration for host-fed input: `slots` in {1,2,3,4} device slots of `slot_bytes`
   each (default 2 x 256 MiB, allocated at the first host feed).  Only between streams. */
int shred_set_ring(shred_ctx *ctx, int slots, uint64_t slot_bytes);

/* Hashing (dedup step 2: "computing a collision-resistant
   hash of the chunk"): SHA-256 (FIPS 180-4; the paper names no function) of every chunk of
   d_in[0..len) delimited by the ascending cuts d_cuts[0 .. *d_ncuts) (e.g. shred_chunk's output,
   chained on the same stream without a host round trip): chunks [0,c0), [c0,c1), ...,
   [c_{n-1}, len), i.e. n+1 chunks (none if len = 0).  d_ncuts is device memory or mapped
   pinned memory; d_cuts must hold all *d_ncuts cuts.  Writes 32 digest bytes per chunk to
   d_digests (16-byte aligned) for at most max_chunks chunks. */
int shred_hash_chunks(shred_ctx *ctx, const uint8_t *d_in, uint64_t len, const uint64_t *d_cuts,
                      const uint64_t *d_ncuts, uint8_t *d_digests, uint64_t max_chunks,
                      shred_stream_t stream);

/* The same for several buffers in one launch sequence (e.g. the files of a backup snapshot,
   PAPER.md L1293-L1361): every buffer's chunks join one length-sorted work list, longest first,
   so the long sequential hash of one buffer's longest chunk overlaps the other buffers' chunks
   instead of idling the GPU (one buffer alone is bound by its longest chunk).  jobs is a HOST
   array of njobs descriptors (each as in shred_hash_chunks; buffers may repeat; digest arrays
   must not overlap); launches take up to 16 jobs at a time. */
typedef struct shred_hash_job {
    const uint8_t *d_in; uint64_t len;
    const uint64_t *d_cuts; const uint64_t *d_ncuts;
    uint8_t *d_digests; uint64_t max_chunks;
} shred_hash_job;
int shred_hash_chunks_batch(shred_ctx *ctx, const shred_hash_job *jobs, int njobs, shred_stream_t stream);

/* Matching (dedup step 3): a device index (hash set) of
   chunk digests owned by the ctx.  shred_index_reset allocates/clears it for `capacity` distinct
   digests (rounded up to a power of two, >= 2x).  shred_index_insert looks up every chunk digest
   produced by shred_hash_chunks (same d_cuts / d_ncuts / len): a chunk is "new" if its digest
   was not in the index (it is then added).  new_flags (optional, device, 1 byte per chunk) gets
   1 for new chunks; the running totals {chunks inserted, new chunks, new bytes, inserts that
   found the index full} are read with shred_index_stats (synchronises).  Of two identical chunks
   inserted by one call exactly one is new. */
int shred_index_reset(shred_ctx *ctx, uint64_t capacity);
int shred_index_insert(shred_ctx *ctx, const uint8_t *d_digests, const uint64_t *d_cuts,
                       const uint64_t *d_ncuts, uint64_t len, uint64_t max_chunks,
                       uint8_t *d_new_flags, shred_stream_t stream);
int shred_index_stats(shred_ctx *ctx, uint64_t stats[4]);

/* Bench/test helper (not the method): writes bytes [offset, offset+len) of the counter-mode
   SplitMix64 stream `seed` into d_buf on `stream`. */
int shred_synth_fill(uint8_t *d_buf, uint64_t len, uint64_t seed, uint64_t offset,
                     shred_stream_t stream);

/* Diagnostics for the bench: kernel launches enqueued by this ctx since creation. */
uint64_t shred_launch_count(const shred_ctx *ctx);

/* Diagnostics for the bench's roofline: while enabled, the ctx records a CUDA event pair on the
   launching stream around every launch of the hot kernel (k1_bulk).  shred_profile_read
   synchronises on the recorded events and returns the summed device time of those launches,
   their number and the input bytes they covered (algorithmic bytes = 1 per input byte), then
   clears the record.  enable = 0 stops recording. */
int shred_profile(shred_ctx *ctx, int enable);

/* Validate *p as shred_init does (no device needed) and report the kernel path an sm_100a
   device runs it on (SHRED_PATH_*) and the hot kernel's marker kind (0: '==' on the low word,
   D = 2^m <= 2^32; 1: '<=' on the low word; 2: '==' by the divisibility test, D = d 2^s with
   s < 32; 3: either marker set on the remainder f - floor(f / D) D, the quotient by a 64-bit
   multiply-high, for every other D).  Either out pointer may be NULL.  SHRED_EINVAL for invalid
   parameters. */
int shred_check_params(const shred_params *p, int *path_out, int *marker_kind_out);

/* Test hook (no device needed): the slot map planning would use for window ends [t_begin, t_end)
   of a job whose bytes start at stream position p_begin at address src_addr, for kernel path
   `path` (SHRED_PATH_*), with (small_ok) or without the small-input launch shape, on sm_count SMs,
   for a window of `window` bytes (1..4096; > 64 never plans a zero lead), zero_lead = 1 if the job starts at the
   stream start with no carried prefix (rows may then start at the stream start itself).
   out[16] = {bulk, small, head_start, head_seg, n_head, b0, S, nrows, tail_start, tail_seg,
   n_tail, bulk CTAs, slot groups, rows per CTA, per-slot list capacity for `divisor`, threads per
   edge CTA}.  SHRED_EINVAL on inconsistent arguments. */
int shred_debug_plan(int path, int small_ok, int sm_count, uint64_t src_addr, uint64_t p_begin,
                     uint64_t t_begin, uint64_t t_end, uint64_t divisor, uint32_t window, int zero_lead,
                     uint64_t out[16]);
/* Test hook (host logic, no GPU): 1 if a multiply-reduction kernel mode applies to poly
   (P = x^k + Q with Q's terms >= 8 apart): K32T for deg <= 32 with the terms below k - 7,
   *mult = Q + 2^k mod 2^32, so T[t] = t(x) x^k mod P ^ (t << k mod 2^32) = t * mult mod 2^32;
   K63T for deg 41..63 with the terms below 25, *mult = Q (low word of T) and
   *mult_hi = 2^(k-32) (high word: the cancel term), so T[t] = (t * mult_hi : t * mult).
   mult / mult_hi may be NULL. */
int shred_debug_tprod(uint64_t poly, uint32_t *mult, uint32_t *mult_hi);
int shred_profile_read(shred_ctx *ctx, double *ms, uint64_t *launches, uint64_t *bytes);

#ifdef __cplusplus
}
#endif
#endif /* SHRED_H */

/*
 * include/jp.h -- C ABI of libjp.so, the B200 (sm_100a) loop-mode engine after
 * Japonica (Han, Zhang, Lam, Wang, ICPP'13).  Citations "P:L<n>" point at
 * /root/reference/PAPER.md lines; "reading Ax" points at DESIGN.md Sec.3.
 *
 * What the library does (P:L17-43 abstract; P:L359-380 and Fig. 2):
 * it executes the iteration space of one annotated loop on the GPU in one of
 * three modes chosen from a profiled dependency density --
 *   DOALL  no cross-iteration dependence,
 *   PRIVATIZED  (private(list) P:L276) only false
 *               (WAR/WAW) dependences, last-writer-wins write-back,
 *   GPU-TLS     (mode B P:L367-375) windowed speculative execution,
 *               RAW check, in-order commit up to the first violator, restart.
 *
 * Conventions (all functions):
 *  - Every pointer is a DEVICE pointer on the current CUDA device unless its
 *    comment says (host).  The caller owns every buffer, including workspace;
 *    the library never allocates device memory and keeps no per-loop state.
 *  - Functions are stream-ordered on `st` and return after enqueueing, EXCEPT
 *    those documented "syncs": they synchronize `st` before returning because
 *    they fill a host struct or must decide a status from device data.
 *  - Errors never abort.  JP_ERR_INDEX (reading A13: an index outside its
 *    array) is detected before any array is modified.  jp_last_error() gives a
 *    thread-local message for the last non-OK status.
 *  - There is no CPU fallback: without a CUDA device every compute entry point
 *    returns JP_ERR_CUDA.
 */
#ifndef JP_H
#define JP_H
#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct CUstream_st *jp_stream_t;   /* == cudaStream_t; NULL = legacy default stream */

typedef enum { JP_OK = 0, JP_ERR_ARG = -1, JP_ERR_CUDA = -2, JP_ERR_WORKSPACE = -3,
               JP_ERR_ILLEGAL_MODE = -4, JP_ERR_INDEX = -5, JP_ERR_UNSUPPORTED = -6 } jp_status;
typedef enum { JP_I32 = 0, JP_F32 = 1 } jp_dtype;
/* The fixed set of templated loop-body opcodes (BASELINE.json north_star).
 * Reads precede writes unless marked "covered".  int32 wraps (reading A11);
 * fp32 is one IEEE RN-even op per operator, never contracted (reading A12).
 *   JP_OP_ADD_C    A[w[i]] = A[r[i]] + c0
 *   JP_OP_SAXPY    Y[w[i]] = c0*X[r[i]] + Y[w[i]]                 (Y in slot A)
 *   JP_OP_PRIV_TMP T[s[i]] = c0*X[r[i]]; Y[w[i]] = T[s[i]] + c1   (T covered; Y in slot A)
 *   JP_OP_STENCIL2 A[w[i]] = (A[r[i]] + A[r2[i]]) * c0           (Gauss-Seidel shape) */
typedef enum { JP_OP_ADD_C = 0, JP_OP_SAXPY = 1, JP_OP_PRIV_TMP = 2, JP_OP_STENCIL2 = 3 } jp_op;
/* Fig. 2(b): A/D' -> DOALL, D -> PRIVATIZED, B -> TLS, C -> SEQ_RECOMMENDED
 * (mode C is "dispatch to CPU"; there is no CPU path, so it is flagged and executed as TLS). */
typedef enum { JP_MODE_DOALL = 0, JP_MODE_PRIVATIZED = 1, JP_MODE_TLS = 2,
               JP_MODE_SEQ_RECOMMENDED = 3 } jp_mode;
/* scheme(s) clause, Table I: sharing (default) or stealing (Sec. V). */
/* JP_SCHED_AUTO: for workflows (jp_schedule_workflow) only -- Sec. V.C. */
typedef enum { JP_SCHED_SHARING = 0, JP_SCHED_STEALING = 1, JP_SCHED_AUTO = 2 } jp_scheme;

typedef union { int32_t i; float f; } jp_scalar;

/* Loop descriptor.  Index arrays are int32 [n]; NULL means identity: local
 * iteration i accesses element ident_off + i.  Element arrays are 4-byte int32
 * or fp32 per `dtype`; A, X, T must not alias each other (reading A14).  Global
 * iteration id of local iteration i is iter_base + i (used by stamps and keys
 * so that chunks/ranks compose); all global ids must be < 2^31 - 1.  A whole
 * loop has iter_base = ident_off = 0; a rank's range [b, e) of a loop over
 * full-size replicas has n = e-b, iter_base = ident_off = b and index arrays
 * offset by b; a range over sharded identity-only arrays keeps ident_off = 0. */
typedef struct {
  int64_t n;                    /* trip count, 0 <= n, iter_base + n <= 2^31-2        */
  int64_t iter_base;            /* global id of local iteration 0                     */
  int64_t ident_off;            /* element index of local iteration 0 under identity  */
  int32_t op;                   /* jp_op                                              */
  int32_t dtype;                /* jp_dtype                                           */
  const int32_t *r, *r2, *w, *s;
  void *A; int64_t len_A;       /* ADD_C/STENCIL2: A;  SAXPY/PRIV_TMP: Y (in/out)     */
  const void *X; int64_t len_X; /* read-only operand (SAXPY, PRIV_TMP)                */
  void *T; int64_t len_T;       /* private(list) scratch, live-out (PRIV_TMP)         */
  jp_scalar c0, c1;
} jp_loop;

/* Dependency density (reading A1; model cited from ref [4]):
 * iteration fractions over the whole loop, any distance, element granularity.
 *   raw_i: an exposed read of i was written by some earlier iteration
 *   war_i: a write of i hits an address read (exposed or covered) earlier
 *   waw_i: a write of i hits an address written earlier                     */
typedef struct {
  int64_t n, raw_iters, war_iters, waw_iters;
  int64_t first_raw_iter;       /* global id, -1 if none                              */
  double d_raw, d_war, d_waw;   /* *_iters / n  (0 when n == 0)                        */
} jp_profile;

typedef struct { int64_t committed, executed, windows, violations; } jp_tls_stats;

/* TLS window policy (reading A8).  window > 0: fixed W.  window == 0: adaptive,
 * W0 = clamp(pow2ceil(ceil(4n/raw)),32,w_max) with a profile (w_max if raw == 0,
 * 4096 without profile), then W <- clamp(pow2ceil(2*max(c,16)), 32, w_max)
 * after a window that committed c iterations.  path: 0 auto (1 when the first
 * window is < 1024 and the window fits, else 3 when it fits a 16-CTA cluster,
 * else 2), 1 single-CTA shared-memory hash path (W <= 4096, 2048 for 3-stream
 * opcodes), 2 cooperative all-SM path (HBM stamps, software grid barrier),
 * 3 one thread-block cluster of `cluster` CTAs (HBM stamps, cluster barriers,
 * W <= 32*(144*cluster - 1)).  cluster: 1..16, 0 = auto (smallest power of two
 * >= 4 that holds the window); ignored by paths 1 and 2.  path 7: no
 * speculation -- one warp runs the loop in program order, 32 iterations per
 * batch, in-batch RAW forwarded by shuffles in dependence order, in-batch WAW
 * resolved to the last writer, the next batch's loads overlapped and patched
 * (mode C, on the device; jp_serial.cu).  Its stats: committed =
 * executed = n, windows = batches, violations = forwarded in-batch reads;
 * window / w_max / cluster / guided / recovery are ignored.                  */
/* Mis-speculation recovery (jp_tls_cfg.recovery).
 * JP_TLS_RESTART (reading A6): commit the prefix before the first violator and
 *   restart the next window there; windows per the policy above.
 * JP_TLS_ONCHIP (reading B7; "commit and mis-speculation recovery",
 *   P:L373-374): fixed windows [kW, (k+1)W); DC finds EVERY violating iteration
 *   of the window, the non-violators commit, and each violator is re-executed
 *   once on chip, in dependence order, with the operand forwarded from its
 *   writer's shadow slot, so every window commits whole.  Needs a profile with
 *   waw_iters == 0 (no address written twice; JP_ERR_ARG otherwise).  window:
 *   fixed W (0 = the largest the path holds); path: 5 one thread-block
 *   cluster, W <= 2048*cluster, cluster 1..16 (0 = auto: the smallest power of
 *   two that holds W, or n when W = 0); 6 every SM (cooperative), W <= 3072 *
 *   co-resident CTAs (454656 on a 148-SM B200, jp_tls_grid_window), write log and shadow values in
 *   workspace regions 7 and 8 (JP_WS_TLS); 8 ONE window of the whole loop
 *   (reading B12; W must be 0 or >= n): ADD_C only, a profile with war_iters ==
 *   waw_iters == 0 and guided = 1 (the guide words of that profile, from
 *   jp_tls_guide or jp_schedule) -- the violators are the guide's raw
 *   iterations, non-violators commit in place at once, violators wait for their
 *   writer's shadow slot (region 8, JP_WS_TLS); no write log, no barrier;
 *   0 = auto (5 when W, or n if W = 0, fits a 16-CTA cluster, else 6; jp_schedule
 *   picks 8 itself when it applies).  w_max is ignored.  stats: windows,
 *   violations = violating iterations, executed = n + violations, committed =
 *   n.  A second writer of an address found at run time (a wrong profile) gives
 *   JP_ERR_ARG after the run, with A in an unspecified state (path 8: a
 *   violator whose writer never published, after a ~seconds-long wait).     */
typedef enum { JP_TLS_RESTART = 0, JP_TLS_ONCHIP = 1 } jp_tls_recovery;
typedef struct {
  int64_t window; int64_t w_max; int32_t path; int32_t cluster;
  int32_t guided;   /* 1: use the guide bitmaps (region 13) that jp_tls_guide wrote for
                       this loop on this workspace; needs a profile with waw_iters == 0
                       (JP_ERR_ARG otherwise).  Same windows, stats and arrays.   */
  int32_t recovery; /* jp_tls_recovery                                          */
} jp_tls_cfg;

typedef struct {
  int32_t scheme;               /* jp_scheme                                          */
  int32_t tls_path;             /* jp_tls_cfg.path                                    */
  double tau_high;              /* Fig. 2(b) "(Density > N)" threshold, reading A4 (0.999, measured) */
  int64_t chunk_iters;          /* task size for stealing / sharing (reading A17)     */
  int64_t tls_window;           /* jp_tls_cfg.window                                  */
  int64_t tls_w_max;            /* jp_tls_cfg.w_max; 0 = auto from the profiled
                                   density: clamp(pow2ceil(sqrt(1000/d_raw)), 256, 1024)
                                   (measured optimum of the single-CTA path)      */
  int32_t tls_recovery;         /* 0 auto (JP_TLS_ONCHIP when the profile shows
                                   waw_iters == 0, else JP_TLS_RESTART -- except
                                   that jp_schedule runs an ADD_C loop with
                                   WAR / WAW profiled by address buckets on path
                                   9 when its last-writer pass holds the loop),
                                   1 restart, 2 on-chip.  With tls_path 0 and tls_recovery 0
                                   a SEQ_RECOMMENDED loop (mode C) runs on the
                                   one-warp program-order path 7              */
  int32_t static_check;         /* 0: before profiling, (a) structural RAW-freedom
                                   (reading B11: PRIV_TMP, and SAXPY with identity
                                   writes, cannot have a true dependence: run
                                   privatized / DOALL after a device check of the
                                   indirect indices, no profile), then (b)
                                   jp_static_check (affine, conflict-free loops
                                   run as DOALL unprofiled); 1: always profile */
} jp_sched_cfg;

typedef struct {
  int32_t mode;                 /* jp_mode of the loop (STEALING: of the first task)  */
  int32_t profiled;             /* 0 when decided statically (all indices NULL,
                                   affine and conflict-free, or reading B11)   */
  jp_profile prof;
  jp_tls_stats tls;
  int64_t n_tasks;              /* STEALING: same-mode chunk runs                     */
  int64_t n_batches;            /* STEALING: topological batches                      */
  int64_t task_mode_iters[4];   /* iterations executed per jp_mode                    */
  int64_t tls_w_max;            /* TLS: the window cap used (auto when cfg 0); the
                                   fixed window under JP_TLS_ONCHIP                */
  int32_t tls_path;             /* TLS: jp_tls_cfg.path that ran (1, 2, 3; 4 tiny
                                   one-CTA schedule; 5 / 6 on-chip recovery on a
                                   cluster / on every SM; 7 one-warp program order
                                   for mode C; 8 on-chip recovery in one window;
                                   9 the same over an ADD_C or SAXPY loop
                                   with WAR / WAW (SAXPY with duplicate
                                   writes: a scatter-add whose writers of one
                                   address chain; reading B14, jp_schedule
                                   only: every
                                   violator fed from the LAST earlier writer of
                                   its address, from a per-iteration shadow slot
                                   in region 8, its index in region 7; last
                                   writers commit at once, or after the window's
                                   one grid barrier when an exposed read of
                                   their address needs the window-start value;
                                   stats as path 8: one window, violations =
                                   raw iterations, jpo_sim_tls_fwd with W = n;
                                   an address with > 4096 writers, or a bucket
                                   of 8192 addresses with > ~49K writes, keeps
                                   the windowed paths))  */
  int32_t tls_guided;           /* TLS: 1 when the guide (jp_tls_guide) steered it    */
  int32_t tls_recovery;         /* TLS: jp_tls_recovery that ran                      */
  int32_t tls_cluster;          /* TLS: CTAs of the cluster (paths 3, 5) or grid (6, 8, 9) */
} jp_sched_result;

/* ---- workspace -------------------------------------------------------------
 * One caller-owned device buffer (256-byte aligned base).  Its regions have
 * FIXED offsets that depend only on the loop (op, which index arrays are NULL,
 * lengths, n), in the order header, profile tables, keys, TLS tables,
 * scheduler scratch; jp_workspace_bytes(L, uses) is the end of the furthest
 * region any of the requested uses (JP_WS_* bits) needs, so a buffer sized for
 * more uses serves every smaller one.  Functions return JP_ERR_WORKSPACE when
 * ws_bytes is too small for what they touch.                                   */
enum { JP_WS_PROFILE = 1, JP_WS_PRIV = 2, JP_WS_TLS = 4, JP_WS_SCHED = 8, JP_WS_GUIDE = 16, JP_WS_ALL = 31 };
size_t jp_workspace_bytes(const jp_loop *L /* host */, int32_t uses);
/* region ids: 0 header, 1 minW(A) int32, 2 minR(A) int32, 3 minW(T), 4 minR(T),
 * 5 keys(A) int64, 6 keys(T) int64, 7 tls stamps(A) u64, 8 tls commit(A) u64,
 * 9 (reserved), 10 tls commit(T) u64 (regions 7 and 8 are the write log S[a] and
 * shadow values V[a] of on-chip TLS recovery on path 6), 11 scheduler scratch, 12 latest exposed
 * reader maxRx(A) int32 (gid, empty -1), 13 TLS guide bitmaps u32 [2][ceil(n/32)]
 * (raw words, then RAW-source words; see jp_tls_guide).  Stamp tables hold
 * INT32_MAX - gid (empty = -1) so that an all_reduce MAX over int32 yields the
 * global first writer/reader; keys hold (gid+1)<<32 | bits32(value) (empty = 0)
 * so that an all_reduce MAX over int64 yields the global last writer.  bytes = 0
 * when the loop does not need the region.  JP_ERR_ARG on a bad id.            */
jp_status jp_ws_region(const jp_loop *L /* host */, int32_t region, size_t *offset /* host */,
                       size_t *bytes /* host */);

/* ---- validation (reading A13) ----------------------------------------------
 * Counts index entries outside their array.  syncs.                          */
jp_status jp_validate(const jp_loop *L, void *ws, size_t ws_bytes, int64_t *bad /* host */,
                      jp_stream_t st);

/* ---- profiler (Fig. 1 "Profiler / DD analysis, intra-warp / inter-warp",
 * P:L127-136) ---------------------------------------------
 * jp_profile_density = jp_profile_stamp + jp_profile_classify.
 * stamp:    clears and fills the first-writer / first-reader tables (regions 1-4)
 *           and validates indices (fused).  Does not sync.
 * classify: per iteration raw/war/waw flags against the tables, counts, optional
 *           raw_bits (uint32[ceil(n/32)], bit i%32 of word i/32 = raw_i) and
 *           optional chunk_counts (int64 [ceil(n/chunk_iters)][3] = raw,war,waw
 *           per chunk of local iterations; chunk_iters % 32 == 0; zeroed by the
 *           call).  syncs; returns JP_ERR_INDEX (nothing modified) if the stamp
 *           pass saw a bad index.                                              */
jp_status jp_profile_stamp(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st);
jp_status jp_profile_classify(const jp_loop *L, void *ws, size_t ws_bytes, uint32_t *raw_bits,
                              int64_t chunk_iters, int64_t *chunk_counts,
                              jp_profile *out /* host */, jp_stream_t st);
jp_status jp_profile_density(const jp_loop *L, void *ws, size_t ws_bytes, uint32_t *raw_bits,
                             int64_t chunk_iters, int64_t *chunk_counts,
                             jp_profile *out /* host */, jp_stream_t st);

/* Fig. 2(b) decision (host only): all index arrays NULL -> DOALL ("determined
 * DOALL"); d_raw > tau_high -> SEQ_RECOMMENDED (mode C); d_raw > 0
 * -> TLS (mode B); d_war > 0 or d_waw > 0 -> PRIVATIZED (mode D); else DOALL
 * (D').  p may be NULL only for the all-NULL case (else JP_ERR_ARG -> -1).   */
int32_t jp_select_mode(const jp_loop *L /* host */, const jp_profile *p /* host, nullable */,
                       double tau_high);

/* ---- static analysis lite (P:L253-256 rule 1, mode A
 * "determined DOALL by static analysis" P:L360-362) -----------------------------
 * One streaming pass decides whether every non-NULL index array is affine in
 * the loop variable (p[i] == alpha*i + beta for all i); NULL arrays are the
 * identity (alpha 1, beta ident_off).  When all are, an exact integer test of
 * every (write, access) pair of the same array (a solution i != j in [0, n) of
 * alpha_f*i + beta_f == alpha_g*j + beta_g) decides `independent`; `in_range`
 * checks every affine index against its array from the endpoints.  syncs.
 * jp_schedule runs it before profiling (jp_sched_cfg.static_check == 0) and
 * executes an independent, in-range loop as DOALL without a profile.       */
typedef struct {
  int32_t affine;               /* 1: every index array is affine                    */
  int32_t independent;          /* 1: affine and free of cross-iteration conflicts   */
  int32_t in_range;             /* 1: affine and every index inside its array        */
  int32_t reserved;
  int64_t alpha[4], beta[4];    /* r, r2, w, s (meaningful when affine)              */
} jp_static;
jp_status jp_static_check(const jp_loop *L, void *ws, size_t ws_bytes, jp_static *out /* host */,
                          jp_stream_t st);
/* The exact test it uses (host only, no device): 1 iff some i != j in [0, n)
 * has af*i + bf == ag*j + bg (|alpha|, |beta| < 2^31, n < 2^31).              */
int32_t jp_affine_dependence(int64_t af, int64_t bf, int64_t ag, int64_t bg, int64_t n);

/* ---- DOALL -------------------------------------------------------
 * Executes all n iterations in place with no protection.  With a profile (host,
 * nullable) that shows any dependence: JP_ERR_ILLEGAL_MODE.  Without a profile
 * the caller asserts legality.  If index arrays are present and p == NULL the
 * indices are validated first (syncs).                                        */
/* Kernel of the affine (all-NULL-index) DOALL body, process-wide: 0 = 16-byte
 * LDG/STG grid-stride stream, 1 = bulk-copy (TMA) staged ring through shared
 * memory (default).  which = 0 or 1 sets it; any other value only queries.
 * Returns the current choice.  Both are bit-exact; DESIGN.md Sec.6 has the
 * measured comparison (initial value from env JP_DOALL_KERNEL).            */
int32_t jp_doall_kernel(int32_t which);
jp_status jp_run_doall(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes,
                       jp_stream_t st);

/* ---- PRIVATIZED, PE(V) (readings A9, A10) -------------
 * Exposed reads see the pre-loop values; covered reads see the iteration's own
 * private copy; every array that some iteration reaches through a non-identity
 * index is written through packed last-writer keys and updated after all
 * iterations; identity-only arrays are stored directly.
 * With a profile showing d_raw > 0: JP_ERR_ILLEGAL_MODE.  Validation as DOALL.
 * Split form for multi-GPU: jp_priv_stream fills the key regions (5, 6; zeroed
 * by the call when `clear_keys`), the caller may all_reduce MAX them, then
 * jp_priv_finalize applies them.                                              */
jp_status jp_run_privatized(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes,
                            jp_stream_t st);
jp_status jp_priv_stream(const jp_loop *L, const jp_profile *p, void *ws, size_t ws_bytes,
                         int32_t clear_keys, jp_stream_t st);
jp_status jp_priv_finalize(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st);

/* ---- GPU-TLS (mode B P:L367-375; readings A6, A7, A8) -------------
 * Windows [ws, we): speculative execution into per-iteration write logs
 * (shadow buffers) with read addresses kept as metadata
 * (P:L326-330); RAW check of every exposed read against earlier in-window
 * writers; commit of the prefix [ws, fv) up to the first violator fv with
 * last-writer-wins; restart at fv.  Always legal.  The whole
 * window loop runs inside one persistent kernel.  stats (host, nullable): if
 * non-NULL the call syncs.  prof (host, nullable) feeds the adaptive policy and
 * lets the commit skip WAW resolution when waw_iters == 0.                   */
/* TLS guide (profile-guided mode B; P:L369-375 uses the
 * profiled density to steer mode B).  From the first-writer table of a
 * jp_profile_stamp on the SAME workspace and loop, fills region 13 with
 *   raw_i = an exposed read of i was written by an earlier iteration, and
 *   src_j = the write of j is an exposed read of some later iteration
 * (a maxRx pass over the exposed reads, region 12).  An in-window RAW
 * violation (reading A7) needs a raw reader and a source writer, so a guided
 * TLS run stamps only sources and checks only raw readers and finds exactly
 * the same first violators.  Needs JP_WS_PROFILE | JP_WS_GUIDE.  No sync.
 * Loops whose A is not reached through an index have no guide (no-op).     */
jp_status jp_tls_guide(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st);
/* Reading A8's adaptive window policy ("sub-loops" of unspecified
 * size), the same function every TLS kernel applies:
 *   prev_commit < 0 (first window): prof_raw_iters < 0 (no profile) -> 4096,
 *     == 0 -> w_max, else pow2ceil(ceil(4n / prof_raw_iters));
 *   after a window that committed c iterations: pow2ceil(2 * max(c, 16));
 * both clamped to [32, w_max].  Host only, no device needed; returns -1 when
 * n < 0 or w_max < 32.                                                       */
int64_t jp_tls_next_window(int64_t n, int64_t prof_raw_iters, int64_t prev_commit, int64_t w_max);
jp_status jp_run_tls(const jp_loop *L, const jp_tls_cfg *cfg /* host */, const jp_profile *prof,
                     void *ws, size_t ws_bytes, jp_tls_stats *stats, jp_stream_t st);

/* ---- scheduler (Sec. V) -----------------------------------------------
 * One GPU, whole loop: static DOALL check, profile, Fig. 2(b) mode, run.
 * scheme STEALING: per-chunk profile; maximal same-mode chunk runs become
 * tasks (Alg. 1 P:L426-437 job pool); tasks that touch a common address with a
 * write are ordered (PDG reading A19), conflict-free tasks of one topological
 * batch run concurrently on separate streams (the TLS task on one SM, the
 * partitioned tasks on the rest).  A SEQ_RECOMMENDED loop (mode C) runs on
 * the one-warp program-order path 7 unless cfg asks for a TLS path or
 * recovery.  The workspace is scratch for the whole call: the profile tables
 * of large loops are kept interleaved in the TLS region and the minW / minR
 * regions are not left filled (call jp_profile_density for the tables).
 * syncs until res is complete (the mode, the profile, the index check); the
 * loop's last writes may still be running on st when it returns (the
 * structurally RAW-free privatized run returns after its index check, before
 * its X -> Y phase; a DOALL exit does not wait at all): read the arrays after
 * st, as for any stream-ordered call.                                      */
jp_status jp_schedule(const jp_loop *L, const jp_sched_cfg *cfg /* host */, void *ws,
                      size_t ws_bytes, jp_sched_result *res /* host */, jp_stream_t st);
/* Same, with every array pointer of L_host on the HOST (pinned for speed): the
 * arrays are copied into `stage` (device, >= jp_stage_bytes), scheduled, and
 * the written arrays copied back.  A determined-DOALL loop (every index NULL,
 * ident_off 0, arrays of n elements) is pipelined instead: chunks of 2^23
 * iterations (env JP_STAGE_CHUNK) go H2D -> kernel -> D2H on three streams, so
 * uploads, kernels and downloads of different chunks overlap (P:L345-349,
 * data staged "asynchronously with the kernel execution"; ws unused).  syncs. */
size_t jp_stage_bytes(const jp_loop *L_host /* host */);
jp_status jp_schedule_host(const jp_loop *L_host /* host */, const jp_sched_cfg *cfg,
                           void *stage, size_t stage_bytes, void *ws, size_t ws_bytes,
                           jp_sched_result *res /* host */, jp_stream_t st);

/* ---- multi-GPU plan (host only; P:L342-358 task sharing, P:L426-460 stealing) ----
 * Task sharing: boundary formula Cg*Fg/(Cg*Fg + Cc*Fc) (garbled at
 * L355; reading A15) generalised to `world` devices with weights[k] = C_k*F_k:
 * rank k gets [floor(n*S_k), floor(n*S_{k+1})) with S_k the prefix sum of the
 * normalised weights (S_world = 1 -> n).  weights NULL = equal.
 * ranges: (host) int64 [world][2].                                            */
jp_status jp_plan_sharing(int64_t n, int32_t world, const double *weights /* host */,
                          int64_t *ranges /* host */);
/* Task stealing (Alg. 1, readings A16, A18) as a deterministic discrete-event
 * plan: tasks (host int64 [n_tasks][3] = start, end, mode) are cut into chunks
 * of chunk_iters (TLS tasks stay whole and pinned to rank 0), dealt to per-rank
 * deques by task sharing, executed head-first at speed[k] iterations per unit
 * time (speed_tls for TLS), and an idle rank steals from the TAIL of the deque
 * with the most remaining iterations (ties: lowest rank).  Output (host):
 * owner[c] for each chunk in order, and n_chunks via *n_out (must be <= cap).  */
jp_status jp_plan_stealing(const int64_t *tasks, int64_t n_tasks, int32_t world,
                           int64_t chunk_iters, const double *speed, double speed_tls,
                           int64_t *chunks /* host [cap][4]: start,end,mode,owner */,
                           int64_t cap, int64_t *n_out, int64_t *stolen_out);

/* ---- workflows: several loops and their PDG (P:L197-200
 * "dependencies between loops are also represented by the program dependency
 * graph", Alg. 1 and P:L438-460 "a task or job refers to a loop and the PDG
 * gives us a workflow", P:L461-469 scheme selection; readings B9, B10) ------
 * Loop u depends on an earlier loop t iff a byte of device memory is written by
 * one of them and read or written by the other (arrays are the ranges
 * [ptr, ptr + 4*len) of A, X, T and the index arrays; A is read by ADD_C,
 * SAXPY and STENCIL2, T and A are written).  batch[u] = 1 + max batch of its
 * dependencies (0 if none): each batch is a set of data-independent loops.
 * scheme AUTO resolves to STEALING when some batch holds >= 2 loops and no
 * loop carries more than half of all iterations ("computations evenly
 * distributed across several data-independent loops"), else SHARING
 * ("heavy computations centralized in only one or few loops").  host only.   */
#define JP_MAX_LOOPS 64
typedef struct {
  int32_t scheme;               /* the scheme the workflow runs with (AUTO resolved) */
  int32_t n_batches;
  int32_t batch[JP_MAX_LOOPS];  /* topological level of each loop                    */
  uint64_t deps[JP_MAX_LOOPS];  /* bit t of deps[u]: loop u depends on loop t < u     */
} jp_workflow_plan;
jp_status jp_plan_workflow(const jp_loop *loops /* host [n] */, int32_t n, int32_t scheme,
                           jp_workflow_plan *out /* host */);
/* Runs a workflow on the current device: SHARING executes the loops in
 * program order, each through jp_schedule with the whole device; STEALING
 * executes batch after batch, the loops of a batch concurrently on separate
 * streams (each through jp_schedule on its own workspace).  cfg->scheme picks
 * the workflow scheme (AUTO allowed); every other cfg field applies to each
 * loop, which runs with the single-loop scheme SHARING.  ws / ws_bytes (host
 * arrays [n]): one workspace per loop (NULL entries: loops that need none).
 * res (host [n]): each loop's jp_sched_result.  syncs.                       */
jp_status jp_schedule_workflow(const jp_loop *loops /* host [n] */, int32_t n, const jp_sched_cfg *cfg,
                               void *const *ws /* host [n] */, const size_t *ws_bytes /* host [n] */,
                               jp_sched_result *res /* host [n] */, jp_workflow_plan *plan /* host */,
                               jp_stream_t st);

/* Apply packed last-writer keys: arr[a] = keys[a] ? lo32(keys[a]) : arr[a]. */
jp_status jp_merge_apply(void *arr, int64_t len, const int64_t *keys, jp_stream_t st);

/* The scheduler's split plan entry (SURVEY §8(b) jp_plan; host only): from
 * per-chunk profiles of the WHOLE loop (chunk_profiles host [n_chunks], chunk
 * k = iterations [k*c, (k+1)*c), c = cfg->chunk_iters or 65536) to per-rank
 * work.  Each chunk gets its Fig. 2(b) mode (cfg->tau_high); maximal runs of
 * one mode are the tasks (reading A19).  cfg->scheme STEALING: the Alg. 1
 * plan of jp_plan_stealing (TLS / mode-C tasks whole and pinned to rank 0,
 * the others cut into chunks, dealt by task sharing, idle ranks stealing
 * tails; speed_tls 1); SHARING: the boundary split of jp_plan_sharing, each
 * rank's range cut at task boundaries.  plan_out (host [plan_cap][4]): rows
 * (start, end, mode, owner); *n_out rows (JP_ERR_ARG with *n_out set when
 * plan_cap is too small).  speed (host [world], nullable): per-rank weights.
 * The inter-task PDG needs the loop's accesses: see jp_plan_tasks.          */
jp_status jp_plan(const jp_loop *L, const jp_sched_cfg *cfg /* host */, const jp_profile *chunk_profiles /* host */,
                  int64_t n_chunks, int32_t world, const double *speed /* host, nullable */,
                  int64_t *plan_out /* host */, int64_t plan_cap, int64_t *n_out /* host */);

/* ---- task stealing across ranks (SURVEY §8(e) "Mixed", Alg. 1) ----
 * The multi-rank stealing scheme (paper_conf_icpp_hanzlw13_b200/dist.py
 * schedule_stealing) needs, on every rank, the same task list and PDG that
 * jp_schedule(STEALING) builds on one device:
 * jp_plan_tasks: chunk_counts (host [3 * ceil(n / chunk_iters)]: raw, war, waw
 * iteration counts of every chunk of the WHOLE loop L, e.g. the sum over the
 * ranks of jp_profile_classify's chunk counts) -> tasks = maximal runs of
 * chunks of one Fig. 2(b) mode (reading A19; SEQ_RECOMMENDED kept as its own
 * mode, run on the one-warp path 7; at most 64, smaller runs merged into the
 * stronger mode, SEQ > TLS > PRIVATIZED > DOALL), tasks (host [3 * 64]) = (start, end, mode) each,
 * *n_tasks; conf (host [64]): bit t of conf[u] set iff tasks t and u touch a
 * common address and at least one writes it (reading B2), computed over L's
 * accesses on this device (workspace JP_WS_ALL of L).  chunk_iters >= 1024, a
 * multiple of 32.  syncs.                                                   */
jp_status jp_plan_tasks(const jp_loop *L, const int64_t *chunk_counts /* host */, int64_t chunk_iters, double tau_high,
                        void *ws, size_t ws_bytes, int64_t *tasks /* host [192] */, int32_t *n_tasks /* host */,
                        uint64_t *conf /* host [64] */, jp_stream_t st);
/* jp_profile_plan_tasks: the same plan from a profile of the WHOLE loop L that
 * this call runs itself (the dependency-density profile of P:L191-196 with
 * per-chunk counts, reading A19; the tasks and PDG of P:L197-200 / P:L441-442,
 * reading B2; every rank holds a full replica: no exchange, identical
 * on every rank) -- by address buckets when L allows it (A >= 2^20, ADD_C /
 * SAXPY; then the task PDG first compares the per-chunk address ranges that
 * profile records), else stamp + classify.  prof (host): the loop's profile;
 * chunk_counts (host [3 * ceil(n / chunk_iters)]): per-chunk raw, war, waw;
 * tasks / n_tasks / conf as jp_plan_tasks.  ws: a workspace of L sized for
 * JP_WS_ALL; its profile, key and scheduler regions are scratch of this call
 * (JP_ERR_WORKSPACE when too small).  JP_ERR_INDEX on an out-of-range index
 * (the loop's arrays are not modified).  syncs.                             */
jp_status jp_profile_plan_tasks(const jp_loop *L, int64_t chunk_iters, double tau_high, void *ws, size_t ws_bytes,
                                jp_profile *prof /* host */, int64_t *chunk_counts /* host */,
                                int64_t *tasks /* host [192] */, int32_t *n_tasks /* host */,
                                uint64_t *conf /* host [64] */, jp_stream_t st);
/* Device-side task stealing of privatized work (Alg. 1: an idle
 * worker steals from the queues of the others).  chunks (device [2 * m]):
 * (start, end) local iterations of L, every chunk free of RAW (a DOALL or
 * PRIVATIZED task's chunks); first (host [world + 1], first[0] = 0): rank k's
 * block of the list is entries [first[k], first[k+1]).  Each rank runs the
 * kernel on its own replica (L, ws): it claims its block's chunks ascending,
 * then the tail of the block with the most unclaimed chunks (ties: lowest
 * rank), with the counter protocol of jp_run_doall_spill (ctr [world] uint64
 * visible to every rank, zero before any rank starts; each chunk runs once).
 * A chunk runs the privatized body: exposed reads see the replica, keyed
 * writes go to ws's key tables by atomicMax (NOT cleared; C4 merges them
 * across ranks afterwards), identity writes are stored in place.  stats
 * (device [3] int64, nullable, accumulated): own iterations, stolen
 * iterations, stolen chunks.  Stream-ordered.                              */
jp_status jp_run_priv_claim(const jp_loop *L, const int64_t *chunks, const int64_t *first /* host [world+1] */,
                            int32_t world, int32_t me, unsigned long long *ctr, int64_t *stats, void *ws,
                            size_t ws_bytes, int32_t max_ctas, jp_stream_t st);
/* Packed last-writer keys (regions keys_A / keys_T of ws, NOT cleared) of what
 * loop L has already written in place: for every iteration i and every
 * indirectly written element a, keys[a] = max(keys[a], (iter_base+i+1) << 32 |
 * bits(current a)).  Used after a TLS task ran in place on its pinned rank so
 * that the other replicas receive its writes through C4 like every privatized
 * task's (reading A9: last writer wins).  Stream-ordered.                   */
jp_status jp_export_keys(const jp_loop *L, void *ws, size_t ws_bytes, jp_stream_t st);

/* ---- task sharing with cross-boundary spill --------
 * the part of the iteration space before the boundary "is divided
 * into uniform chunks of moderate size, which are executed ... in an ascending
 * order, while the right part is executed ... in a descending order"; the two
 * consumers meet wherever the faster one gets to.  Generalised to k ranks:
 * rank k's range (its task-sharing share, jp_plan_sharing) is cut into
 * ceil(n_k / chunk) chunks; rank k consumes its own chunks ascending and, once
 * they are all claimed, takes chunks DESCENDING from the tail of the rank with
 * the most unclaimed chunks (ties: lowest rank; reading A18).
 *
 * views (host [world], world <= 8): every rank's shard as a loop descriptor
 * whose pointers are valid in THIS process (the caller maps peer shards, e.g.
 * with jp_ipc_import; on one device they are plain pointers).  Affine shards
 * only: all index arrays NULL, ident_off 0, the same op / dtype / c0 / c1.
 * ctr (device [world] uint64, visible to every rank, zero before ANY rank
 * starts): ctr[k] = (tail claims << 32) | head claims of rank k's chunks,
 * advanced with one system-scope atomicAdd per claim, so every chunk runs
 * exactly once whatever the interleaving.  stats (device [3] int64, nullable,
 * accumulated: the caller zeroes): iterations of own chunks, iterations
 * stolen, chunks stolen by this executor.  max_ctas > 0 caps the grid.
 * Results are complete when EVERY rank's launch has finished (the caller
 * synchronises and barriers).  Stream-ordered.                               */
jp_status jp_run_doall_spill(const jp_loop *views /* host [world] */, int32_t world, int32_t me, int64_t chunk,
                             unsigned long long *ctr, int64_t *stats, int32_t max_ctas, jp_stream_t st);
/* C4 over NVLink peer memory, for small key tables (len <= 16384, e.g. config
 * 4's 1024 private slots; SURVEY §2c C9's role without NCCL).  Every rank calls
 * it once per merge, after its privatized stream on the same stream:
 * peer_keys (host [world]): every rank's key table (this rank's included) as
 * device pointers valid here (jp_ipc_import); keys: this rank's table; bar: a
 * uint64 counter visible to every rank (in one rank's memory), zero before the
 * first call and never reset; epoch: 1, 2, ... (the same on every rank).  One
 * CTA per rank: a device-side barrier (system-scope atomicAdd + acquire
 * polling of bar) until every rank's keys are in, the max of every slot over
 * the ranks, a second barrier until every rank has read, then keys = the
 * merged table and, when arr is not NULL, arr[a] = lo32(keys[a]) where
 * keys[a] != 0 (jp_merge_apply's rule, reading A9).  A barrier waiting over
 * ~4 s sets *err (device int32, caller zeroes) to 1 and abandons the merge.
 * Stream-ordered.                                                          */
jp_status jp_keys_merge_p2p(const int64_t *const *peer_keys /* host [world] */, int32_t world, int64_t *keys,
                            int64_t len, unsigned long long *bar, int64_t epoch, void *arr, int32_t *err,
                            jp_stream_t st);
/* Privatized stream + C4 + R2 in ONE kernel per rank (config-4 shape: PRIV_TMP,
 * identity X / Y, indirect s, len_T <= 4096; SURVEY Sec.8(e) "C4 ... or inside
 * the kernel"; the paper updates privatized variables "after all the iterations
 * finish execution", reading A9).  L is this rank's range
 * (iter_base = global id of its first iteration).  After every CTA's key flush
 * and a grid barrier, one CTA pushes this rank's len_T packed keys into slot
 * (epoch parity, me) of EVERY rank's inbox (plain stores to peer memory over
 * NVLink), raises one release flag per peer, waits for all world flags of this
 * epoch in its own inbox, reduces the world tables (MAX, local loads) and
 * applies the last writers to T.  inbox: jp_priv_inbox_bytes bytes per rank,
 * zeroed once before the first call; peer_inbox (host [world]) holds every
 * rank's inbox pointer as mapped in this process (own included; CUDA IPC).
 * The epoch lives in the inbox, so the call's launches (a key memset and one
 * cooperative kernel) take the same arguments every step: a CUDA graph can
 * capture them.  Every rank calls it once per step; a wait over ~4 s sets *err
 * (device int32, caller zeroes) to 1 and leaves T unmerged.  Stream-ordered.   */
size_t jp_priv_inbox_bytes(const jp_loop *L /* host */, int32_t world);
jp_status jp_priv_stream_merge(const jp_loop *L, const jp_profile *p /* host, nullable */, void *ws, size_t ws_bytes,
                               void *const *peer_inbox /* host [world] */, int32_t world, int32_t me,
                               int32_t *err, jp_stream_t st);
/* CUDA IPC plumbing for the spill (peer shards and the counter table):
 * export: a 64-byte handle (host) of the allocation holding ptr, and ptr's
 * byte offset in it; import (in another process): *ptr = mapped base + offset
 * (peer access enabled lazily); close: unmap what import returned.           */
jp_status jp_ipc_export(const void *ptr, void *handle /* host, 64 B */, int64_t *offset /* host */);
jp_status jp_ipc_import(const void *handle /* host, 64 B */, int64_t offset, void **ptr /* host */);
jp_status jp_ipc_close(void *ptr, int64_t offset);

/* ---- owner-partitioned sparse exchange --------
 * Building blocks for the "one exchange step" of partitioned loops with
 * indirect writes: the whole-loop first-writer / first-reader tables of the
 * profile (reading A1; C1) and the last-writer keys of the privatized write-
 * back (reading A9; C4) are per-address MAX reductions over the
 * ranks.  Instead of all-reducing the dense tables, a rank packs the entries
 * it touched into rows bucketed by the address's OWNER rank
 * (owner(a) = a / ceil(len / world)), the caller all_to_alls them, and the
 * owner folds them into its slice (the library never calls NCCL).
 *
 * A table is a dense device array of len elements of elem_bytes: 4 (int32,
 * compared signed; len <= INT32_MAX) or 8 (uint64, compared unsigned).  One or
 * two tables of the same length travel together (t1 NULL: one).  A row is
 * 1 + ntab elements of elem_bytes, row-major: column 0 the address, then the
 * value of each table at that address.                                       */

/* Scratch (device, caller-owned, 8-byte aligned) jp_sparse_pack needs.       */
size_t jp_sparse_scratch_bytes(int64_t len, int32_t world);
/* Rows for every address a in [lo, hi) where t0[a] != empty or
 * t1[a] != empty, in increasing address order -- hence grouped by owner --
 * written to rows[0 .. m) (m = sum of counts).  counts (host [world]):
 * number of rows of each owner (owners computed over the whole [0, len)).
 * cap: capacity of rows in rows; when m > cap nothing beyond cap is written
 * and JP_ERR_ARG is returned with counts filled.  syncs.                     */
jp_status jp_sparse_pack(const void *t0, const void *t1 /* nullable */, int32_t elem_bytes, int64_t len,
                         int64_t lo, int64_t hi, int64_t empty, int32_t world, void *rows, int64_t cap,
                         int64_t *counts /* host [world] */, void *scratch, size_t scratch_bytes, jp_stream_t st);
/* For each of the m rows: t_q[addr] = max(t_q[addr], row value q), atomic,
 * in any order (MAX is order-free).  Rows with addr outside [0, len) are
 * ignored (padding).                                                          */
jp_status jp_sparse_reduce_max(void *t0, void *t1 /* nullable */, int32_t elem_bytes, int64_t len, const void *rows,
                               int64_t m, jp_stream_t st);
/* For each row (in place): row value q = t_q[addr]; out-of-range rows are left as they are. */
jp_status jp_sparse_gather(const void *t0, const void *t1 /* nullable */, int32_t elem_bytes, int64_t len, void *rows,
                           int64_t m, jp_stream_t st);
/* For each row: t_q[addr] = row value q.  Rows must carry distinct addresses
 * (as pack produces them; otherwise which row lands is unspecified);
 * out-of-range rows are ignored.                                              */
jp_status jp_sparse_scatter(void *t0, void *t1 /* nullable */, int32_t elem_bytes, int64_t len, const void *rows,
                            int64_t m, jp_stream_t st);

const char *jp_last_error(void);
const char *jp_version(void);
/* Number of kernels this library has launched in this process (for bench.py). */
int64_t jp_launch_count(void);
/* The largest window of on-chip TLS path 6 on the current device (co-resident
 * CTAs x 512 threads x 6 slots: 454656 on a 148-SM B200); 0 without a device. */
int64_t jp_tls_grid_window(void);

#ifdef __cplusplus
}
#endif
#endif /* JP_H */

// jp_host.h -- host-side internals of libjp.so (workspace layout, launchers).
#pragma once
#include <cstddef>
#include <cstdint>
#include <cuda_runtime.h>
#include "jp_internal.cuh"

namespace jp {

enum Region : int {
  R_HEADER = 0, R_MINW_A = 1, R_MINR_A = 2, R_MINW_T = 3, R_MINR_T = 4, R_KEYS_A = 5,
  R_KEYS_T = 6, R_TLS_S_A = 7, R_TLS_C_A = 8, R_TLS_S_T = 9, R_TLS_C_T = 10, R_SCHED = 11,
  R_MAXRX_A = 12, R_GUIDE = 13, R_COUNT = 14
};

struct Layout {
  size_t off[R_COUNT];
  size_t bytes[R_COUNT];
  size_t total;
};

// cudaFuncSetAttribute(fn, MaxDynamicSharedMemorySize, bytes) once per (kernel,
// device) and size: the attribute call costs about a microsecond of host time on
// every launch otherwise (the launch-bound front of jp_schedule)
cudaError_t set_smem_once(const void *fn, int bytes);
// host-side phase marks (JP_HOST_TRACE=1: microseconds since the previous mark, to stderr)
void htrace(const char *what);

// Fixed-offset layout of a workspace for loop L (offsets do not depend on uses).
Layout layout(const jp_loop *L);
// End of the furthest region the JP_WS_* uses touch.
size_t layout_end(const Layout &lo, int uses);
constexpr int64_t kSchedMinChunk = 1024;
// Reading A4's threshold of Fig. 2(b) "(Density > N)", measured: the
// one-window on-chip TLS beats the one-warp program-order path (mode C) on every
// loop of the crossover sweep up to d_raw = 0.999 (chains, delta = 1: 131 vs 19 M
// committed iter/s at 0.999; 0.88 vs 18.95 at 1.0), so mode C starts above 0.999
// (bench.py modes.crossover, profiles/r02_bench.json; DESIGN.md Sec.3 A4)
constexpr double kTauHigh = 0.999;
constexpr int kMaxTasks = 64;
// scheduler scratch sub-layout (inside R_SCHED)
struct SchedLayout {
  size_t counts, chunk_task, wmA, rmA, wmT, rmT, conf, tstats, ranges, crange, total;
};
SchedLayout sched_layout(const jp_loop *L);

template <typename T> inline T *at(void *ws, const Layout &lo, int r) {
  return lo.bytes[r] ? reinterpret_cast<T *>(static_cast<char *>(ws) + lo.off[r]) : nullptr;
}

// A (sub-)loop ready to launch: the device view plus its opcode and dtype.
struct Job {
  DLoop d;
  int op, dt;
};
Job make_job(const jp_loop *L);

// ---- launchers (each returns the first CUDA error, if any) ----
cudaError_t launch_validate(const Job &j, int64_t *hdr, cudaStream_t st);
// the index arrays reached through an index (identity accesses are checked on the
// host by check_loop) against their lengths: *bad = number out of range; no sync
cudaError_t launch_validate_indirect(const Job &j, int64_t *bad, cudaStream_t st);
// TLS guide bitmaps (region R_GUIDE: raw words then source words) from the
// stamp tables of a profile on the same workspace; no sync.
cudaError_t launch_tls_guide(const Job &j, void *ws, const Layout &lo, cudaStream_t st);
// pairs: stamp the A tables into interleaved {minW, minR} pairs in region 7 (see stamp_pairs_ok)
cudaError_t launch_prof_stamp(const Job &j, void *ws, const Layout &lo, cudaStream_t st, bool pairs = false,
                              bool pairs_ready = false);
bool stamp_pairs_ok(const Job &j, void *ws, const Layout &lo);
// the profile by address buckets (jp_bucket.cu): counts, first raw, raw-distance
// histogram, optional guide words (zeroed here) and per-chunk counts, for ADD_C /
// SAXPY loops over a large A; uses minW/minR_A and maxRx_A as scratch (their
// tables are NOT left filled).  bucket_profile_ok says whether it applies.
bool bucket_profile_ok(const Job &j, void *ws, const Layout &lo);
// one-window on-chip TLS (path 8, jp_tls_flow.cu): ADD_C loops with a profile
// showing waw = war = 0 and the guide words of that profile; stats as noted there
// wsrc (nullable) with lo: a range [lo, lo + n) of a loop whose profile recorded the
// writer of every raw read (loop-local ids, wsrc indexed by the range's local i):
// a raw read whose writer precedes the range reads A (committed) and is no violator
// gate (nullable): a profile header the kernel checks before running (launched
// ahead of the host's read of it): it exits at once unless H_BAD = H_WAR =
// H_WAW = 0 and 0 < H_RAW <= raw_max
cudaError_t launch_tls_flow(const Job &j, const uint32_t *graw, const uint32_t *gsrc, unsigned long long *V,
                            int64_t *stats, cudaStream_t st, const int32_t *wsrc = nullptr, int64_t lo = 0,
                            const int64_t *gate = nullptr, int64_t raw_max = 0, bool zero_stats = true,
                            int max_ctas = 0, uint32_t *o = nullptr, int64_t ph_max = 0);
// (o, n words of scratch, with a gate: when the gate's raw count is at most ph_max
// the non-violators' values are gathered by a kernel of their own first and the
// sweep only scatters them -- JP_FLOW_PHASED=0 keeps the one-kernel form)
// wsrc (nullable, ADD_C): the first writer of every raw iteration's read (int32 [n])
// crange (nullable, needs chunk % 16384 == 0): per chunk the min and max address of A
// the chunk touches (uint32 [2 * chunks]) -- the stealing scheduler's task ranges
// vclr (nullable, ADD_C): V[a] = 0 at the address of every raw read -- every slot
// the one-window TLS (path 8) polls or publishes, so V needs no full clear
// sample_m > 0: the first kernel also runs the static check's affine sample on
// the first sample_m entries of every index array (verdict to hdr[H_GATE] and to
// the mapped host words mir[0], then seq to mir[1]); when the sample looks
// affine every later kernel of the profile exits at once (H_GATE = 1), so the
// host can queue the whole profile before it knows the verdict
cudaError_t launch_prof_bucket(const Job &j, void *ws, const Layout &lo, uint32_t *graw, uint32_t *gsrc,
                               int64_t chunk, int64_t *cc, cudaStream_t st, int32_t *wsrc = nullptr,
                               uint32_t *crange = nullptr, unsigned long long *vclr = nullptr, int sample_m = 0,
                               long long *mir = nullptr, const unsigned long long *seq = nullptr);
// (seq: a mapped host word holding the call's sequence number, written by the
// host before the launch -- the launches are replayed from a CUDA graph per
// argument set, JP_NO_GRAPHS=1 issues them one by one)
constexpr int64_t kBucketTile = 16384;   // (jp_bucket.cu's tile: chunk ranges need chunk % kBucketTile == 0)
// after launch_prof_bucket on the same workspace (its records still in place),
// ADD_C: the last earlier writer of every raw read -> pred[i] (raw i only), and
// three bitmaps of nw = ceil(n/32) words at bits (zeroed here): publish (the
// writer is some raw read's pred), now (last writer of an address no exposed read
// touches), later (last writer of an address that has an exposed read).
// hdr[H_PRED_FAIL] > 0 if the pass could not hold some bucket's writers.  V[pred]
// = 0 for every pred (the only per-iteration shadow slots path 9 polls).
cudaError_t launch_prof_pred(const Job &j, void *ws, const Layout &lo, int32_t *pred, uint32_t *bits,
                             unsigned long long *V, cudaStream_t st);
// one-window on-chip TLS over a loop with WAR / WAW (path 9, reading B14): pred and
// bits from launch_prof_pred, graw the profile's raw words, V one tagged shadow
// slot per ITERATION (V[pred] zeroed by launch_prof_pred); the kernel exits at once
// if gate[H_PRED_FAIL] != 0.
// stats as launch_tls_flow's (stats[3] violations, stats[1] lost warps)
cudaError_t launch_tls_flow_waw(const Job &j, const uint32_t *graw, const int32_t *pred, const uint32_t *bits,
                                unsigned long long *V, int64_t *stats, const int64_t *gate, cudaStream_t st);
// src_bits (nullable): also the TLS guide's RAW-source words (raw_bits then holds its raw words)
cudaError_t launch_prof_classify(const Job &j, void *ws, const Layout &lo, uint32_t *raw_bits,
                                 int64_t chunk, int64_t *chunk_counts, cudaStream_t st, uint32_t *src_bits = nullptr,
                                 bool stamped_pairs = false);
// counts + the TLS guide bitmaps (region 13, valid when the loop writes no address twice) in one pass
cudaError_t launch_prof_classify_guide(const Job &j, void *ws, const Layout &lo, cudaStream_t st,
                                       bool stamped_pairs = false);
// o (nullable, n words of scratch): an indirect loop other than PRIV_TMP runs as a
// gather kernel (every iteration's value into o) then a scatter kernel
// (JP_DOALL_PHASED=0 keeps the one-kernel form)
cudaError_t launch_doall(const Job &j, cudaStream_t st, int max_ctas = 0, uint32_t *o = nullptr);
int doall_kernel_choice();
void set_doall_kernel_choice(int v);
// fuse_apply: the stream kernel may also apply the keys (single-GPU PE(V));
// *applied tells whether it did (then launch_priv_finalize is not needed)
// validate (nullable): count out-of-range indirect indices into *validate before
// anything is written (reading A13; j.d.abort should point at it so that every
// later kernel of the run exits when it is nonzero)
// mirror (nullable, mapped host words): the two-phase kernel (fused apply with
// validate) writes mirror[0] = the count, then mirror[1] = seq, as soon as the
// check is done; *published tells whether that kernel ran (else read *validate)
cudaError_t launch_priv_stream(const Job &j, void *ws, const Layout &lo, bool clear_keys,
                               cudaStream_t st, int max_ctas = 0, bool fuse_apply = false, bool *applied = nullptr,
                               int64_t *validate = nullptr, int64_t *mirror = nullptr, unsigned long long seq = 0,
                               bool *published = nullptr);
cudaError_t launch_priv_finalize(const Job &j, void *ws, const Layout &lo, cudaStream_t st);
cudaError_t launch_merge_apply(void *arr, int64_t len, const int64_t *keys, cudaStream_t st);
// mode C on the device (jp_serial.cu): one warp runs the loop in program order; stats[4] as TLS
cudaError_t launch_serial(const Job &j, int64_t *stats, cudaStream_t st);
// device-side task stealing of privatized chunks (Alg. 1), keys to regions 5/6
cudaError_t launch_priv_claim(const Job &j, void *ws, const Layout &lo, const int64_t *chunks, const int64_t *first,
                              int world, int me, unsigned long long *ctr, int64_t *stats, int max_ctas,
                              cudaStream_t st);
// the privatized stream of a config-4-shaped rank range with C4 over peer memory and
// R2 fused into its epilogue (jp_priv_stream_merge); inbox = every rank's inbox mapped here
bool priv_merge_ok(const Job &j, int world);
size_t priv_inbox_bytes(const Job &j, int world);
cudaError_t launch_priv_stream_merge(const Job &j, unsigned long long *kT, unsigned long long *const *inbox, int world,
                                     int me, int *err, cudaStream_t st);
// C4 over NVLink peer memory: merged max of every rank's key table (len <= kP2PMaxLen), applied to arr
constexpr int64_t kP2PMaxLen = 16384;
cudaError_t launch_keys_merge_p2p(const unsigned long long *const *peers, int world, unsigned long long *mine,
                                  int64_t len, unsigned long long *bar, unsigned long long epoch, uint32_t *arr,
                                  int *err, cudaStream_t st);
// keys (regions 5/6) of what loop j already wrote in place (atomicMax, keys not cleared)
cudaError_t launch_export_keys(const Job &j, void *ws, const Layout &lo, cudaStream_t st);
// task sharing with cross-boundary spill (jp_doall.cu, C8): views[k] = rank k's affine shard
constexpr int kSpillRanks = 8;
cudaError_t launch_doall_spill(const Job *views, int world, int me, int64_t chunk, unsigned long long *ctr,
                               int64_t *stats, int max_ctas, cudaStream_t st);
// owner-partitioned sparse exchange (jp_exchange.cu)
size_t sparse_scratch_bytes(int64_t len, int world);
int64_t sparse_pack_tiles(int64_t len, int64_t lo, int64_t hi, int world);
cudaError_t launch_sparse_pack(const void *t0, const void *t1, int elem, int64_t len, int64_t lo, int64_t hi,
                               int64_t empty, int world, void *rows, int64_t cap, int64_t *counts_dev, void *scratch,
                               cudaStream_t st);
// what: 0 reduce max, 1 gather, 2 scatter
cudaError_t launch_sparse_rows(void *t0, void *t1, int elem, int64_t len, void *rows, int64_t m, int what,
                               cudaStream_t st);
// STEALING scheduler helpers (jp_sched.cu): per-task write/read bitmasks of every
// address, then the task x task conflict matrix conf[t] (bit u set: t and u
// touch a common address and at least one of them writes it).
// per-task address ranges rg [4][kMaxTasks] uint32 (minA, maxA, minT, maxT; empty: min > max)
cudaError_t launch_task_ranges(const Job &j, const int32_t *chunk_task, int64_t chunk, uint32_t *rg, cudaStream_t st);
cudaError_t launch_task_conflicts(const Job &j, const int32_t *chunk_task, int64_t chunk, int n_tasks,
                                  unsigned long long *wmA, unsigned long long *rmA,
                                  unsigned long long *wmT, unsigned long long *rmT,
                                  unsigned long long *conf, cudaStream_t st);

// static analysis lite (jp_static.cu): flags[q] = index array q (r, r2, w, s) is affine
cudaError_t launch_affine(const Job &j, int *flags, cudaStream_t st);
// one warp: mir[0] = 1 when the first m (>= 2) entries of every index array are
// affine, then mir[1] = seq (mapped host words, st.release.sys)
cudaError_t launch_prefix_affine(const Job &j, int m, long long *mir, unsigned long long seq, cudaStream_t st);
bool affine_conflict(int64_t af, int64_t bf, int64_t ag, int64_t bg, int64_t n);

// tiny loops (jp_tiny.cu): the whole schedule in one CTA's shared memory
bool tiny_eligible(const jp_loop *L);
// mirror (nullable, mapped pinned host [17]): header words 0..15 then seq, written by the kernel
cudaError_t launch_tiny(const Job &j, const jp_loop *L, double tau, int64_t window, int64_t w_max, int recovery,
                        int64_t *hdr, cudaStream_t st, int64_t *mirror = nullptr, unsigned long long seq = 0);

struct TlsPlan {
  int64_t window, w_max, prof_raw;  // prof_raw < 0: no profile
  bool waw;                         // in-window WAW resolution needed
  int path;                         // 1 cta, 2 grid, 3 cluster, 5 on-chip recovery cluster
  int cluster;                      // CTAs of the cluster paths (power of two)
  bool guided;                      // stamp only RAW sources, check only RAW readers
  int recovery;                     // jp_tls_recovery
};
// on-chip recovery path (jp_tls_fwd.cu, reading B7): fixed window (> 0), cluster of C CTAs
// bits / bsrc: guide words (raw readers / RAW sources) of local iteration 0's word, or NULL (unguided)
cudaError_t launch_tls_fwd(const Job &j, int64_t window, int cluster, const uint32_t *bits, const uint32_t *bsrc,
                           int64_t *stats, cudaStream_t st);
int64_t tls_fwd_wcap(int cluster);   // largest window a C-CTA cluster holds (2048*C)
int tls_fwd_max_cluster();           // 16 when the device schedules it, else 8
// on-chip recovery over every SM (cooperative): S, V = u64 [lenS] (regions 7, 8), bar = 2 zeroed u32
cudaError_t launch_tls_fwd_grid(const Job &j, int64_t window, const uint32_t *bits, const uint32_t *bsrc,
                                unsigned long long *S,
                                unsigned long long *V, int64_t lenS, unsigned *bar, int64_t *stats,
                                cudaStream_t st, int clean = 0);   // bit 0: S clean, bit 1: V zeroed
int64_t tls_fwd_grid_wcap();         // slots per CTA * co-resident CTAs (2048 * 148 on B200)
int64_t tls_fwd_grid_cta_slots();    // window iterations per CTA of the all-SM kernel
// stats: int64[4] device (committed, executed, windows, violations); bar: u32[2]
// zeroed barrier words + int64[3] fv slots (grid path).
cudaError_t launch_tls(const Job &j, void *ws, const Layout &lo, const TlsPlan &p, int64_t *stats,
                       cudaStream_t st);
int64_t tls_next_window(int64_t n, int64_t prof_raw, int64_t prev_commit, int64_t w_max);
int64_t tls_cluster_wcap(int cluster);
int64_t tls_cta_wcap(int op, bool waw, bool guided);   // largest single-CTA window
int tls_max_cluster();                                 // 16 when the device schedules it, else 8
#ifdef JP_TLS_TRACE
cudaError_t tls_trace_copy(long long *host, int n);
cudaError_t tls_fwd_trace_copy(long long *host, int n);
#endif

}  // namespace jp

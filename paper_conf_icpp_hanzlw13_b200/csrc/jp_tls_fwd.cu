// jp_tls_fwd.cu -- GPU-TLS with on-chip mis-speculation recovery (DESIGN.md
// reading B7, mode B P:L367-375).
//
// The paper's sub-loop goes through "speculative execution (SE), dependency
// checking (DC), commit and mis-speculation recovery"; DC tells
// "which threads fell in violation" and the threads "not found to
// have violations" commit; violating warps are re-run
// "sequentially".  The classic path (jp_tls.cu) commits the prefix
// before the first violator and restarts the window there (reading A6).  This
// path keeps the whole window on chip instead and recovers the violators in
// place: every iteration speculates against the memory of the window start
// (its write goes to a shadow slot, never to A), DC looks every exposed read
// up in the window's write log, and a violating iteration is re-executed once,
// in dependence order, with the operand forwarded from its writer's shadow slot
// -- so each window ends in the sequential state and commits whole.  Legal when
// no address is written twice (profile waw_iters == 0): then an exposed read's
// in-window earlier writer is unique and its shadow value is exactly what the
// sequential loop would read.
//
// One thread-block cluster of C CTAs (C <= 16) runs the window loop; window
// offset off = k*G + g (G = C*512 threads, g = the thread's cluster-wide id,
// k < 4 slots), so the window holds up to 2048*C iterations.
//   write log  an open-addressing hash of (address, writer offset) spread over
//              the C CTAs' shared memory (slot s lives in CTA s >> 12), three
//              tables used round-robin so a table is cleared one window after
//              its last reader and one window before its next writer; inserts
//              and probes are DSMEM CAS / loads.
//   shadow     OV[k*512 + t] in the owning CTA: (epoch << 32 | value); a
//              re-executing violator polls its writer's slot until the epoch
//              matches (writers are always earlier, so the wait chain ends).
//   pipeline   ONE cluster barrier per window.  The next window's gathers are
//              issued right after it (they see every earlier window's commit)
//              and the current window's own writes are forwarded into them at
//              the end of the window from the write log.
//   stats      windows, violations (violating iterations), executed = n +
//              violations (one re-execution each), committed = n -- the
//              definition of oracle/jpo.c jpo_sim_tls_fwd.
// Guided (jp_tls_guide bitmaps): only RAW-source writes are logged and only
// raw readers probe the log or take forwarded values -- the same violators.
#include <cstdio>
#include "jp_host.h"
#include "jp_internal.cuh"

namespace jp {

constexpr int kFwdThreads = 512;
constexpr int kFwdK = 4;                       // window slots per thread
constexpr int kFwdHashLog = 12;                // write-log slots per CTA per table
constexpr int kFwdHash = 1 << kFwdHashLog;
constexpr int kFwdTables = 3;
constexpr uint32_t kNone = 0xFFFFFFFFu;
constexpr unsigned long long kFwdEmpty = ~0ull;
constexpr size_t kFwdSmem = (size_t)kFwdTables * kFwdHash * 8 + (size_t)kFwdK * kFwdThreads * 8;

int64_t tls_fwd_wcap(int cluster) { return (int64_t)kFwdThreads * kFwdK * cluster; }

__device__ __forceinline__ uint32_t fwd_rank() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
  return r;
}
__device__ __forceinline__ void fwd_cluster_sync() {
  asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
__device__ __forceinline__ uint32_t dsm_map(uint32_t local, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(local), "r"(rank));
  return r;
}
__device__ __forceinline__ unsigned long long dsm_ld(uint32_t a) {
  unsigned long long v;
  asm volatile("ld.relaxed.cluster.shared::cluster.u64 %0, [%1];" : "=l"(v) : "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ void dsm_st(uint32_t a, unsigned long long v) {
  asm volatile("st.relaxed.cluster.shared::cluster.u64 [%0], %1;" ::"r"(a), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long dsm_cas(uint32_t a, unsigned long long cmp, unsigned long long v) {
  unsigned long long old;
  asm volatile("atom.relaxed.cluster.shared::cluster.cas.b64 %0, [%1], %2, %3;" : "=l"(old) : "r"(a), "l"(cmp), "l"(v)
               : "memory");
  return old;
}
__device__ __forceinline__ void dsm_red_add(uint32_t a, uint32_t v) {
  asm volatile("red.relaxed.cluster.shared::cluster.add.u32 [%0], %1;" ::"r"(a), "r"(v) : "memory");
}

// the write log: C * kFwdHash slots per table, slot s in CTA s >> kFwdHashLog
struct FwdLog {
  uint32_t base;     // shared address of this CTA's tables
  int logTot;        // log2(C * kFwdHash)
  __device__ __forceinline__ uint32_t home(uint32_t key) const { return (key * 0x9E3779B1u) >> (32 - logTot); }
  __device__ __forceinline__ uint32_t addr(int tab, uint32_t s) const {
    return dsm_map(base + (((uint32_t)tab << kFwdHashLog) + (s & (kFwdHash - 1))) * 8u, s >> kFwdHashLog);
  }
  // claim a slot for (key, off); returns the slot, or kNone when the key is
  // already logged in this window (a second writer: WAW, flagged by the caller)
  __device__ __forceinline__ uint32_t insert(int tab, uint32_t key, uint32_t off) const {
    const unsigned long long mine = ((unsigned long long)key << 32) | off;
    const uint32_t mask = (1u << logTot) - 1;
    uint32_t s = home(key);
    while (true) {
      const unsigned long long old = dsm_cas(addr(tab, s), kFwdEmpty, mine);
      if (old == kFwdEmpty) return s;
      if ((uint32_t)(old >> 32) == key) return kNone;
      s = (s + 1) & mask;
    }
  }
  // writer offset of key in the window, kNone if none
  __device__ __forceinline__ uint32_t find(int tab, uint32_t key) const {
    const uint32_t mask = (1u << logTot) - 1;
    uint32_t s = home(key);
    while (true) {
      const unsigned long long v = dsm_ld(addr(tab, s));
      if ((uint32_t)(v >> 32) == key) return (uint32_t)v;
      if (v == kFwdEmpty) return kNone;
      s = (s + 1) & mask;
    }
  }
};

// values of one iteration from its two operands (see the opcode table, include/jp.h)
template <int OP, int DT>
__device__ __forceinline__ uint32_t fwd_body(const DLoop &L, uint32_t a0, uint32_t a1, uint32_t &vt) {
  if constexpr (OP == JP_OP_ADD_C) return op_add<DT>(a0, L.c0);
  else if constexpr (OP == JP_OP_SAXPY) return op_add<DT>(op_mul<DT>(L.c0, a0), a1);
  else if constexpr (OP == JP_OP_PRIV_TMP) { vt = op_mul<DT>(L.c0, a0); return op_add<DT>(vt, L.c1); }
  else return op_mul<DT>(op_add<DT>(a0, a1), L.c0);
}

template <int OP, int DT, bool GUIDED>
__global__ void __launch_bounds__(kFwdThreads, 1)
    k_tls_fwd(DLoop L, int track, int logC, uint32_t W, const uint32_t *graw, const uint32_t *gsrc, int64_t *stats) {
  constexpr int T = kFwdThreads, K = kFwdK;
  // ops whose exposed A read may hit another iteration's write: ADD_C A[r],
  // STENCIL2 A[r], A[r2].  SAXPY reads Y[w] (its own write address) and X;
  // PRIV_TMP reads X: with no address written twice they never violate.
  constexpr bool kTr = OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2;
  constexpr bool k2 = OP == JP_OP_STENCIL2;
  extern __shared__ __align__(16) unsigned long long fsm[];
  unsigned long long *OV = fsm + kFwdTables * kFwdHash;   // [K][T] shadow slots
  __shared__ uint32_t s_cnt[2];                            // violations, duplicate writers (CTA 0's are the totals)
  const uint32_t crank = fwd_rank();
  const int tid = threadIdx.x;
  const uint32_t G = (uint32_t)T << logC;
  const uint32_t g = crank * T + (uint32_t)tid;
  const uint32_t n32 = (uint32_t)L.n;
  const uint32_t io = (uint32_t)L.ioff;
  const bool trk = kTr && track;
  FwdLog H{smem_u32(fsm), kFwdHashLog + logC};
  const uint32_t ovbase = smem_u32(OV);

  for (int k = tid; k < kFwdTables * kFwdHash; k += T) fsm[k] = kFwdEmpty;
  for (int k = tid; k < K * T; k += T) OV[k] = 0;   // epoch 0: never published
  if (tid == 0) { s_cnt[0] = 0; s_cnt[1] = 0; }
  fwd_cluster_sync();

  // shadow slot of window offset j: CTA (j % G) / T, local (j / G) * T + j % T
  auto ov_addr = [&](uint32_t j) {
    const uint32_t gj = j & (G - 1);
    return dsm_map(ovbase + (((j >> (9 + logC)) << 9) + (gj & (T - 1))) * 8u, gj >> 9);
  };

  int32_t cr[K], cw[K], c2[K];      // indices of the current window (r, w, r2 or s)
  int32_t nr[K], nw[K], n2[K];      // indices of the next window
  uint32_t cb = 0, nb = 0;          // guide bits: bit k raw_i, bit K+k src_i
  uint32_t g0[K], g1[K];            // operands of the current window (window-start values)
  uint32_t ng0[K], ng1[K];          // gathered operands of the next window
  uint32_t ins[K], pins[K];         // write-log slots inserted in this / the previous window

  auto load_idx = [&](uint32_t ws, int32_t *R, int32_t *Wi, int32_t *R2, uint32_t &bits) {
    bits = 0;
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g, i = ws + off;
      if (off < W && i < n32) {
        R[k] = L.r ? __ldg(L.r + i) : (int32_t)(io + i);
        Wi[k] = L.w ? __ldg(L.w + i) : (int32_t)(io + i);
        if constexpr (OP == JP_OP_STENCIL2) R2[k] = L.r2 ? __ldg(L.r2 + i) : (int32_t)(io + i);
        if constexpr (OP == JP_OP_PRIV_TMP) R2[k] = L.s ? __ldg(L.s + i) : (int32_t)(io + i);
        if constexpr (GUIDED) {
          bits |= ((__ldg(graw + (i >> 5)) >> (i & 31)) & 1u) << k;
          bits |= ((__ldg(gsrc + (i >> 5)) >> (i & 31)) & 1u) << (K + k);
        }
      }
    }
  };
  auto gather = [&](uint32_t ws, const int32_t *R, const int32_t *Wi, const int32_t *R2, uint32_t *a0, uint32_t *a1) {
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g;
      if (off < W && ws + off < n32) {
        if constexpr (OP == JP_OP_ADD_C) a0[k] = __ldcg(L.A + R[k]);
        else if constexpr (OP == JP_OP_SAXPY) { a0[k] = __ldg(L.X + R[k]); a1[k] = __ldcg(L.A + Wi[k]); }
        else if constexpr (OP == JP_OP_PRIV_TMP) a0[k] = __ldg(L.X + R[k]);
        else { a0[k] = __ldcg(L.A + R[k]); a1[k] = __ldcg(L.A + R2[k]); }
      }
    }
  };

  const uint32_t nwin = (n32 + W - 1) / W;
  load_idx(0, cr, cw, c2, cb);
  gather(0, cr, cw, c2, g0, g1);
  if (nwin > 1) load_idx(W, nr, nw, n2, nb);
#pragma unroll
  for (int k = 0; k < K; k++) { ins[k] = kNone; pins[k] = kNone; }
  uint32_t viol = 0, dup = 0;
  int tab = 0;

  for (uint32_t win = 0; win < nwin; win++) {
    const uint32_t ws = win * W, epoch = win + 1;
    const bool more = win + 1 < nwin;
    // ---------------- SE: log this window's writes ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g;
      ins[k] = kNone;
      const bool act = off < W && ws + off < n32;
      bool log = trk && act;
      if constexpr (GUIDED) log = log && ((cb >> (K + k)) & 1u);
      if (log) {
        ins[k] = H.insert(tab, (uint32_t)cw[k], off);
        dup += ins[k] == kNone;
      }
    }
    fwd_cluster_sync();   // the write log is complete; earlier windows' commits are visible
    // the previous window's table is no longer read by anyone: clear my slots of it
    const int ptab = tab == 0 ? kFwdTables - 1 : tab - 1;
#pragma unroll
    for (int k = 0; k < K; k++)
      if (pins[k] != kNone) dsm_st(H.addr(ptab, pins[k]), kFwdEmpty);
    // next window's operands (this window's own writes are forwarded into them below)
    if (more) gather(ws + W, nr, nw, n2, ng0, ng1);
    // ---------------- DC: every exposed read against the window's write log ----------------
    uint32_t src0[K], src1[K];
    uint32_t pend = 0;
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g;
      src0[k] = src1[k] = kNone;
      const bool act = off < W && ws + off < n32;
      bool chk = trk && act;
      if constexpr (GUIDED) chk = chk && ((cb >> k) & 1u);
      if (chk) {
        const uint32_t j0 = H.find(tab, (uint32_t)cr[k]);
        if (j0 < off) src0[k] = j0;
        if constexpr (k2) {
          const uint32_t j1 = H.find(tab, (uint32_t)c2[k]);
          if (j1 < off) src1[k] = j1;
        }
      }
      if (src0[k] != kNone || src1[k] != kNone) pend |= 1u << k;
    }
    viol += __popc(pend);
    // ---------------- speculative values of the non-violators -> shadow slots ----------------
    uint32_t va[K], vt[K];
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g;
      if (off < W && ws + off < n32 && !((pend >> k) & 1u)) {
        va[k] = fwd_body<OP, DT>(L, g0[k], g1[k], vt[k]);
        *(volatile unsigned long long *)&OV[k * T + tid] = ((unsigned long long)epoch << 32) | va[k];
      }
    }
    // ---------------- recovery: violators re-execute with forwarded operands ----------------
    while (__any_sync(0xffffffffu, pend)) {
#pragma unroll
      for (int k = 0; k < K; k++) {
        if ((pend >> k) & 1u) {
          bool ready = true;
          uint32_t a0 = g0[k], a1 = g1[k];
          if (src0[k] != kNone) {
            const unsigned long long v = dsm_ld(ov_addr(src0[k]));
            if ((uint32_t)(v >> 32) == epoch) a0 = (uint32_t)v; else ready = false;
          }
          if constexpr (k2) {
            if (src1[k] != kNone) {
              const unsigned long long v = dsm_ld(ov_addr(src1[k]));
              if ((uint32_t)(v >> 32) == epoch) a1 = (uint32_t)v; else ready = false;
            }
          }
          if (ready) {
            va[k] = fwd_body<OP, DT>(L, a0, a1, vt[k]);
            *(volatile unsigned long long *)&OV[k * T + tid] = ((unsigned long long)epoch << 32) | va[k];
            pend &= ~(1u << k);
          }
        }
      }
    }
    // ---------------- commit: the whole window ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g;
      if (off < W && ws + off < n32) {
        __stcg(L.A + cw[k], va[k]);
        if constexpr (OP == JP_OP_PRIV_TMP) __stcg(L.T + c2[k], vt[k]);
      }
    }
    // ---------------- forward this window's writes into the next window's operands ----------------
    uint32_t fx = 0, f0[K], f1[K];
    if (more && trk) {
#pragma unroll
      for (int k = 0; k < K; k++) {
        const uint32_t off = (uint32_t)k * G + g;
        bool chk = off < W && ws + W + off < n32;
        if constexpr (GUIDED) chk = chk && ((nb >> k) & 1u);
        if (chk) {
          const uint32_t j0 = H.find(tab, (uint32_t)nr[k]);
          if (j0 != kNone) {
            unsigned long long v;
            do { v = dsm_ld(ov_addr(j0)); } while ((uint32_t)(v >> 32) != epoch);
            f0[k] = (uint32_t)v;
            fx |= 1u << k;
          }
          if constexpr (k2) {
            const uint32_t j1 = H.find(tab, (uint32_t)n2[k]);
            if (j1 != kNone) {
              unsigned long long v;
              do { v = dsm_ld(ov_addr(j1)); } while ((uint32_t)(v >> 32) != epoch);
              f1[k] = (uint32_t)v;
              fx |= 1u << (K + k);
            }
          }
        }
      }
    }
    // ---------------- rotate ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      cr[k] = nr[k]; cw[k] = nw[k];
      if constexpr (OP == JP_OP_STENCIL2 || OP == JP_OP_PRIV_TMP) c2[k] = n2[k];
      g0[k] = ((fx >> k) & 1u) ? f0[k] : ng0[k];
      g1[k] = ((fx >> (K + k)) & 1u) ? f1[k] : ng1[k];
      pins[k] = ins[k];
    }
    cb = nb;
    if (win + 2 < nwin) load_idx(ws + 2 * W, nr, nw, n2, nb);
    tab = tab == kFwdTables - 1 ? 0 : tab + 1;
  }
  // ---------------- stats (CTA 0 sums the cluster) ----------------
  viol = __reduce_add_sync(0xffffffffu, viol);
  dup = __reduce_add_sync(0xffffffffu, dup);
  if ((tid & 31) == 0 && (viol | dup)) {
    const uint32_t a = dsm_map(smem_u32(s_cnt), 0);
    if (viol) dsm_red_add(a, viol);
    if (dup) dsm_red_add(a + 4, dup);
  }
  fwd_cluster_sync();
  if (crank == 0 && tid == 0) {
    const int64_t v = *(volatile uint32_t *)&s_cnt[0];
    stats[0] = s_cnt[1] ? -1 : (int64_t)n32;   // -1: a second writer of an address (caller's profile was wrong)
    stats[1] = (int64_t)n32 + v;
    stats[2] = nwin;
    stats[3] = v;
  }
}

// ---------------------------------------------------------------------------
// grid path: every SM.  The window holds up to 2048 * CTAs iterations; the
// write log is a stamp table S[a] = epoch << 32 | writer offset and the shadow
// slots are V[a] = epoch << 32 | value, both in global memory (L2) and indexed
// by ADDRESS (an address has at most one writer in the loop, so neither is
// ever cleared: a stale epoch reads as "no writer in this window").  A reader
// that finds an earlier in-window writer in S polls V at its own read address.
// One software grid barrier per window (monotone counter, release/acquire).
// ---------------------------------------------------------------------------
__device__ __forceinline__ void fwd_grid_sync(unsigned *count, unsigned target) {
  JP_CTA_SYNC();
  if (threadIdx.x == 0) {
    asm volatile("fence.acq_rel.gpu;\n\tred.relaxed.gpu.global.add.u32 [%0], 1;" ::"l"(count) : "memory");
    unsigned v;
    do {
      asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(count) : "memory");
    } while (v < target);
    asm volatile("fence.acq_rel.gpu;" ::: "memory");
  }
  JP_CTA_SYNC();
}
__device__ __forceinline__ unsigned long long g_ld_relaxed(const unsigned long long *p) {
  unsigned long long v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void g_st_relaxed(unsigned long long *p, unsigned long long v) {
  asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}

// Per-window state of one thread: the indices, guide bits and operands of its
// K slots.  The kernel keeps two of these and alternates them (a two-window
// unrolled loop), so loads issued for the next window land in registers that
// are not touched again until that window runs: no register copy ever waits
// on an outstanding load.
template <int K>
struct FwdSet {
  int32_t r[K], w[K], x[K];   // read / write / (r2 | s) addresses
  uint32_t g0[K], g1[K];      // operands (window-start values, patched by forwarding)
  uint32_t gr[K], gs[K];      // guide words holding the slot's raw-reader / RAW-source bit (read
                              // where the bit is used, so the loads never stall the index prefetch)
};

#ifdef JP_TLS_TRACE
// phase marks (SM clock) of CTA 0 / thread 0 per window (trace build only, scripts/tls_fwd_trace.py)
__device__ long long g_fwd_trace[2048 * 16];
cudaError_t tls_fwd_trace_copy(long long *host, int n) {
  return cudaMemcpyFromSymbol(host, g_fwd_trace, sizeof(long long) * (size_t)n);
}
#define FTR(ph) do { if (blockIdx.x == 0 && threadIdx.x == 0 && win < 2048u) g_fwd_trace[win * 16 + (ph)] = clock64(); } while (0)
#else
#define FTR(ph) do { } while (0)
#endif

// the all-SM kernel's CTA shape (threads x window slots per thread); the
// window is 148 x kGridT x kGridK iterations
#ifndef JP_GRID_T
#define JP_GRID_T 512
#endif
#ifndef JP_GRID_K
#define JP_GRID_K 6
#endif
constexpr int kGridT = JP_GRID_T, kGridK = JP_GRID_K;
#ifndef JP_GRID_EARLY_GATHER
#define JP_GRID_EARLY_GATHER 0
#endif

template <int OP, int DT, bool GUIDED, int K>
struct FwdGrid {
  static constexpr bool kTr = OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2;
  static constexpr bool k2 = OP == JP_OP_STENCIL2;
  static constexpr int T = kGridT;
  DLoop L;
  const uint32_t *graw, *gsrc;
  unsigned long long *S, *V;
  unsigned *bar;
  uint32_t W, G, g, n32, io, nwin;
  bool trk;
  uint32_t viol = 0, dup = 0;

  __device__ __forceinline__ bool act(uint32_t ws, int k) const {
    const uint32_t off = (uint32_t)k * G + g;
    return off < W && ws + off < n32;
  }
  __device__ __forceinline__ void load_idx(uint32_t ws, FwdSet<K> &s) const {
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (!act(ws, k)) continue;
      // streamed once: evict-first, so that the gathered array stays in L2
      const uint32_t i = ws + (uint32_t)k * G + g;
      s.r[k] = L.r ? __ldcs(L.r + i) : (int32_t)(io + i);
      s.w[k] = L.w ? __ldcs(L.w + i) : (int32_t)(io + i);
      if constexpr (OP == JP_OP_STENCIL2) s.x[k] = L.r2 ? __ldcs(L.r2 + i) : (int32_t)(io + i);
      if constexpr (OP == JP_OP_PRIV_TMP) s.x[k] = L.s ? __ldcs(L.s + i) : (int32_t)(io + i);
      if constexpr (GUIDED) {
        s.gr[k] = __ldcs(graw + (i >> 5));
        s.gs[k] = __ldcs(gsrc + (i >> 5));
      }
    }
  }
  // gathers of a window's operands; skip: bit k = operand 0 of slot k already
  // forwarded, bit K+k = operand 1
  __device__ __forceinline__ void gather(uint32_t ws, FwdSet<K> &s, uint32_t skip = 0) const {
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (!act(ws, k)) continue;
      const bool s0 = (skip >> k) & 1u, s1 = (skip >> (K + k)) & 1u;
      if constexpr (OP == JP_OP_ADD_C) { if (!s0) s.g0[k] = __ldcg(L.A + s.r[k]); }
      else if constexpr (OP == JP_OP_SAXPY) { s.g0[k] = __ldg(L.X + s.r[k]); s.g1[k] = __ldcg(L.A + s.w[k]); }
      else if constexpr (OP == JP_OP_PRIV_TMP) s.g0[k] = __ldg(L.X + s.r[k]);
      else { if (!s0) s.g0[k] = __ldcg(L.A + s.r[k]); if (!s1) s.g1[k] = __ldcg(L.A + s.x[k]); }
    }
  }
  // guide bits of slot k of the window starting at ws (true when unguided)
  __device__ __forceinline__ bool raw_bit(const FwdSet<K> &s, uint32_t ws, int k) const {
    if constexpr (GUIDED) return (s.gr[k] >> ((ws + (uint32_t)k * G + g) & 31)) & 1u;
    else return true;
  }
  __device__ __forceinline__ bool src_bit(const FwdSet<K> &s, uint32_t ws, int k) const {
    if constexpr (GUIDED) return (s.gs[k] >> ((ws + (uint32_t)k * G + g) & 31)) & 1u;
    else return true;
  }
  static __device__ __forceinline__ bool cur(unsigned long long v, unsigned long long tag) {
    return (v & ~0xFFFFFFFFull) == tag;
  }

  // one window: c = this window's set (indices, operands), nx = the next window's
  // set (indices loaded; its gathers are issued here; its indices for the window
  // after it are loaded into c at the end)
  __device__ __forceinline__ void step(uint32_t win, FwdSet<K> &c, FwdSet<K> &nx) {
    const uint32_t ws = win * W, epoch = win + 1;
    const unsigned long long tag = (unsigned long long)epoch << 32;
    const bool more = win + 1 < nwin;
    FTR(0);
    // ---------------- SE: log this window's writes (S[w] = epoch | offset) ----------------
    unsigned long long old[K];
#pragma unroll
    for (int k = 0; k < K; k++) {
      old[k] = 0;
      if (trk && act(ws, k) && src_bit(c, ws, k)) old[k] = atomicExch(S + c.w[k], tag | ((uint32_t)k * G + g));
    }
    FTR(1);
    fwd_grid_sync(bar, gridDim.x * epoch);
    FTR(2);
#if JP_GRID_EARLY_GATHER
    // the next window's gathers right after the barrier, so their latency hides
    // behind this window's DC / publish / commit; operands this window writes
    // are stale here and are replaced below by forwarding (a read of an element
    // written in this window is a raw read, hence probed: q0 / q1)
    if (more) gather(ws + W, nx, 0);
#endif
    // ---------------- this window's DC probes and the next window's forwarding
    // probes, all at once; the next window's gathers wait for the end of the
    // window so that probes and polls do not queue behind them ----------------
    unsigned long long p0[K], p1[K], q0[K], q1[K];
#pragma unroll
    for (int k = 0; k < K; k++) {
      p0[k] = p1[k] = q0[k] = q1[k] = 0;
      if (trk && act(ws, k) && raw_bit(c, ws, k)) {
        p0[k] = __ldcg(S + c.r[k]);
        if constexpr (k2) p1[k] = __ldcg(S + c.x[k]);
      }
      if (trk && more && act(ws + W, k) && raw_bit(nx, ws + W, k)) {
        q0[k] = __ldcg(S + nx.r[k]);
        if constexpr (k2) q1[k] = __ldcg(S + nx.x[k]);
      }
    }
    // ---------------- DC ----------------
    uint32_t pend = 0;   // bit k: operand 0 of slot k waits for its writer; bit K+k: operand 1
#pragma unroll
    for (int k = 0; k < K; k++) {
      const uint32_t off = (uint32_t)k * G + g;
      if (cur(p0[k], tag) && (uint32_t)p0[k] < off) pend |= 1u << k;
      if constexpr (k2) if (cur(p1[k], tag) && (uint32_t)p1[k] < off) pend |= 1u << (K + k);
    }
    viol += __popc((pend | (pend >> K)) & ((1u << K) - 1));
    FTR(3);
    // ---------------- non-violators: values, published where a later reader may wait ----------------
    uint32_t va[K], vt[K];
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (act(ws, k) && !(((pend >> k) | (pend >> (K + k))) & 1u)) {
        va[k] = fwd_body<OP, DT>(L, c.g0[k], c.g1[k], vt[k]);
        if (trk && src_bit(c, ws, k)) g_st_relaxed(V + c.w[k], tag | va[k]);
      }
    }
    FTR(4);
    // ---------------- recovery ----------------
#ifdef JP_TLS_TRACE
    int npass = 0;
    const bool anyp = __any_sync(0xffffffffu, pend);
    FTR(9);
    if (blockIdx.x == 0 && threadIdx.x == 0 && win < 2048u) g_fwd_trace[win * 16 + 11] = anyp;
#endif
    while (__any_sync(0xffffffffu, pend)) {
#ifdef JP_TLS_TRACE
      npass++;
#endif
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (((pend >> k) | (pend >> (K + k))) & 1u) {
          if ((pend >> k) & 1u) {
            const unsigned long long v = g_ld_relaxed(V + c.r[k]);
            if (cur(v, tag)) { c.g0[k] = (uint32_t)v; pend &= ~(1u << k); }
          }
          if constexpr (k2) {
            if ((pend >> (K + k)) & 1u) {
              const unsigned long long v = g_ld_relaxed(V + c.x[k]);
              if (cur(v, tag)) { c.g1[k] = (uint32_t)v; pend &= ~(1u << (K + k)); }
            }
          }
          if (!(((pend >> k) | (pend >> (K + k))) & 1u)) {
            va[k] = fwd_body<OP, DT>(L, c.g0[k], c.g1[k], vt[k]);
            if (src_bit(c, ws, k)) g_st_relaxed(V + c.w[k], tag | va[k]);
          }
        }
      }
    }
    FTR(5);
#ifdef JP_TLS_TRACE
    if (blockIdx.x == 0 && threadIdx.x == 0 && win < 2048u) g_fwd_trace[win * 16 + 10] = npass;
#endif
    // ---------------- commit ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (act(ws, k)) {
        __stcg(L.A + c.w[k], va[k]);
        if constexpr (OP == JP_OP_PRIV_TMP) __stcg(L.T + c.x[k], vt[k]);
      }
    }
    FTR(6);
    // ---------------- forward this window's writes into the next window's operands,
    // then gather the rest of them ----------------
    uint32_t fwd = 0;
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (cur(q0[k], tag)) {
        unsigned long long v;
        do { v = g_ld_relaxed(V + nx.r[k]); } while (!cur(v, tag));
        nx.g0[k] = (uint32_t)v;
        fwd |= 1u << k;
      }
      if constexpr (k2) {
        if (cur(q1[k], tag)) {
          unsigned long long v;
          do { v = g_ld_relaxed(V + nx.x[k]); } while (!cur(v, tag));
          nx.g1[k] = (uint32_t)v;
          fwd |= 1u << (K + k);
        }
      }
    }
#if !JP_GRID_EARLY_GATHER
    if (more) gather(ws + W, nx, fwd);
#endif
    // a second writer of an address in this window (checked last: the log
    // atomics' return values must not hold up the probes issued after the barrier)
#pragma unroll
    for (int k = 0; k < K; k++) dup += (uint32_t)(old[k] >> 32) == epoch;
    FTR(7);
    if (win + 2 < nwin) load_idx(ws + 2 * W, c);
    FTR(8);
  }
};

template <int OP, int DT, bool GUIDED>
__global__ void __launch_bounds__(kGridT, 1)
    k_tls_fwd_grid(DLoop L, int track, uint32_t W, const uint32_t *graw, const uint32_t *gsrc, unsigned long long *S,
                   unsigned long long *V, unsigned *bar, int64_t *stats) {
  constexpr int K = kGridK;
  FwdGrid<OP, DT, GUIDED, K> F;
  F.L = L; F.graw = graw; F.gsrc = gsrc; F.S = S; F.V = V; F.bar = bar;
  F.W = W;
  F.G = gridDim.x * (uint32_t)kGridT;
  F.g = blockIdx.x * (uint32_t)kGridT + threadIdx.x;
  F.n32 = (uint32_t)L.n;
  F.io = (uint32_t)L.ioff;
  F.nwin = (F.n32 + W - 1) / W;
  F.trk = FwdGrid<OP, DT, GUIDED, K>::kTr && track;
  FwdSet<K> A, B;
  F.load_idx(0, A);
  F.gather(0, A);
  if (F.nwin > 1) F.load_idx(W, B);
  for (uint32_t win = 0; win < F.nwin; win += 2) {
    F.step(win, A, B);
    if (win + 1 < F.nwin) F.step(win + 1, B, A);
  }
  // ---------------- stats: stats[3] and the dup counter (bar[1]) were zeroed by the launcher ----------------
  const int tid = threadIdx.x;
  uint32_t viol = __reduce_add_sync(0xffffffffu, F.viol);
  uint32_t dup = __reduce_add_sync(0xffffffffu, F.dup);
  if ((tid & 31) == 0) {
    if (viol) atomicAdd(reinterpret_cast<unsigned long long *>(&stats[3]), (unsigned long long)viol);
    if (dup) atomicAdd(bar + 1, dup);
  }
  fwd_grid_sync(bar, gridDim.x * (F.nwin + 1));
  if (blockIdx.x == 0 && tid == 0) {
    const int64_t v = *(volatile int64_t *)&stats[3];
    stats[0] = *(volatile unsigned *)(bar + 1) ? -1 : (int64_t)F.n32;
    stats[1] = (int64_t)F.n32 + v;
    stats[2] = F.nwin;
  }
}

template <int OP, int DT>
static void run_fwd_grid(cudaError_t &e, const Job &j, uint32_t W, const uint32_t *bits, const uint32_t *bsrc,
                         unsigned long long *S,
                         unsigned long long *V, unsigned *bar, int64_t *stats, cudaStream_t st) {
  void *fn = bits ? (void *)k_tls_fwd_grid<OP, DT, true> : (void *)k_tls_fwd_grid<OP, DT, false>;
  const int grid = (int)((W + kGridT * kGridK - 1) / (kGridT * kGridK));
  int maxb = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&maxb, fn, kGridT, 0);
  if (grid > num_sms() * (maxb > 0 ? maxb : 1)) { e = cudaErrorInvalidConfiguration; return; }
  DLoop d = j.d;
  int track = a_indirect(j.op, j.d.r, j.d.r2, j.d.w) ? 1 : 0;
  void *args[] = {&d, &track, &W, &bits, &bsrc, &S, &V, &bar, &stats};
  e = cudaLaunchCooperativeKernel(fn, dim3(grid), dim3(kGridT), args, 0, st);
  note_launch();
}

cudaError_t launch_tls_fwd_grid(const Job &j, int64_t window, const uint32_t *bits, const uint32_t *bsrc,
                                unsigned long long *S,
                                unsigned long long *V, int64_t lenS, unsigned *bar, int64_t *stats,
                                cudaStream_t st, int clean) {
  if (j.d.n == 0) {
    cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
    return launch_check();
  }
  if (S && lenS > 0) {   // epoch 0: no writer yet
    // clean bit 0: S holds this call's {minW, minR} stamp pairs, whose high words
    // (encoded gids >= 2^31 - 2^24, or all ones) never equal a window epoch
    // (< 2^24): they already read as "no writer this window"
    // clean bit 1: the caller already zeroed V (on a side stream, behind the profile)
    if (!(clean & 1)) cudaMemsetAsync(S, 0, 8 * (size_t)lenS, st);
    if (!(clean & 2)) cudaMemsetAsync(V, 0, 8 * (size_t)lenS, st);
  }
  cudaMemsetAsync(bar, 0, 2 * sizeof(unsigned), st);
  cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
  cudaError_t e = cudaSuccess;
  JP_DISPATCH(j.op, j.dt, run_fwd_grid, e, j, (uint32_t)window, bits, bsrc, S, V, bar, stats, st);
  if (e != cudaSuccess) return e;
  return launch_check();
}

int64_t tls_fwd_grid_cta_slots() { return (int64_t)kGridT * kGridK; }

int64_t tls_fwd_grid_wcap() {
  int maxb = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&maxb, (void *)k_tls_fwd_grid<JP_OP_ADD_C, JP_I32, true>, kGridT, 0);
  cudaGetLastError();
  return (int64_t)kGridT * kGridK * num_sms() * (maxb > 0 ? maxb : 1);
}

// Largest cluster (power of two <= 16) the device schedules for k_tls_fwd (cached per device).
int tls_fwd_max_cluster() {
  static int cache[64] = {0};
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= 64) return 8;
  if (cache[dev]) return cache[dev];
  int best = 8;
  void *fn = (void *)k_tls_fwd<JP_OP_ADD_C, JP_I32, true>;
  if (cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1) == cudaSuccess &&
      cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)kFwdSmem) == cudaSuccess) {
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(16, 1, 1);
    cfg.blockDim = dim3(kFwdThreads, 1, 1);
    cfg.dynamicSmemBytes = kFwdSmem;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeClusterDimension;
    attr[0].val.clusterDim.x = 16;
    attr[0].val.clusterDim.y = 1;
    attr[0].val.clusterDim.z = 1;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    int n = 0;
    if (cudaOccupancyMaxActiveClusters(&n, fn, &cfg) == cudaSuccess && n >= 1) best = 16;
  }
  cudaGetLastError();
  cache[dev] = best;
  return best;
}

template <int OP, int DT>
static void run_fwd(cudaError_t &e, const Job &j, uint32_t W, int C, const uint32_t *bits, const uint32_t *bsrc,
                    int64_t *stats, cudaStream_t st) {
  int logC = 0;
  while ((1 << logC) < C) logC++;
  void *fn = bits ? (void *)k_tls_fwd<OP, DT, true> : (void *)k_tls_fwd<OP, DT, false>;
  e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)kFwdSmem);
  if (e != cudaSuccess) return;
  if (C > 8 && (e = cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1)) != cudaSuccess) return;
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3(C, 1, 1);
  cfg.blockDim = dim3(kFwdThreads, 1, 1);
  cfg.dynamicSmemBytes = kFwdSmem;
  cfg.stream = st;
  cudaLaunchAttribute attr[1];
  attr[0].id = cudaLaunchAttributeClusterDimension;
  attr[0].val.clusterDim.x = C;
  attr[0].val.clusterDim.y = 1;
  attr[0].val.clusterDim.z = 1;
  cfg.attrs = attr;
  cfg.numAttrs = 1;
  DLoop d = j.d;
  int track = a_indirect(j.op, j.d.r, j.d.r2, j.d.w) ? 1 : 0;
  void *args[] = {&d, &track, &logC, &W, &bits, &bsrc, &stats};
  e = cudaLaunchKernelExC(&cfg, fn, args);
  note_launch();
}

cudaError_t launch_tls_fwd(const Job &j, int64_t window, int cluster, const uint32_t *bits, const uint32_t *bsrc,
                           int64_t *stats, cudaStream_t st) {
  if (j.d.n == 0) {
    cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
    return launch_check();
  }
  cudaError_t e = cudaSuccess;
  JP_DISPATCH(j.op, j.dt, run_fwd, e, j, (uint32_t)window, cluster, bits, bsrc, stats, st);
  if (e != cudaSuccess) return e;
  return launch_check();
}

}  // namespace jp

// jp_tiny.cu -- the whole scheduler for tiny loops in one CTA (config 1:
// N = 4096, |A| = 4096).  jp_schedule on such a loop would otherwise cost ~8
// API calls and two host synchronisations around microseconds of work; here
// one launch does profile (P1/P2, reading A1) -> Fig. 2(b) mode (P:L399-416,
// reading A4/A5) -> the chosen mode, with the in/out arrays, the index
// streams and every table staged in shared memory, then one D2H of the
// results.  Semantics are those of the large-loop kernels (same readings):
//   DOALL       in place, any order (legal: no dependence at all);
//   PRIVATIZED  exposed reads from the pre-loop snapshot, covered T reads from
//               the iteration's own value, last writer per address wins (A9, A10);
//   TLS         prefix-commit windows (A6, A7) with the adaptive policy A8;
//               write stamps direct-mapped per address (the address space is
//               small): S[a] = (kTinyEpochs - epoch) << 12 | offset, atomicMin,
//               so a newer window's stamp always wins over a stale one; the
//               commit order per address is a second table, atomicMax of
//               epoch << 13 | offset + 1 (last committed writer wins).
#include <cmath>
#include "jp_host.h"

namespace jp {

constexpr int kTinyThreads = 1024, kTinyK = 4;   // n <= 4096 (few warps: everything is in shared memory)
constexpr uint32_t kTinyEpochs = 0xFFFFF;        // 20-bit window counter (windows <= n <= 4096)

struct TinyArgs {
  double tau;
  int64_t window, w_max;   // w_max 0: from the profiled density (as jp_schedule)
  int recovery;            // jp_sched_cfg.tls_recovery: 0 auto (on chip when no address is written twice), 1 restart
  int64_t *mirror;         // nullable: mapped pinned host words [17] = header words 0..15, then seq
  unsigned long long seq;
};

// the result words straight into mapped host memory, then the sequence flag:
// the host polls the flag instead of enqueueing a D2H copy (config 1 is
// launch-latency bound).  Every thread's stores are fenced before the flag.
__device__ __forceinline__ void tiny_publish(const int64_t *hdr, const TinyArgs &a) {
  if (!a.mirror) return;
  __threadfence();
  JP_CTA_SYNC();
  if (threadIdx.x == 0) {
    for (int k = 0; k < 16; k++) a.mirror[k] = hdr[k];
    __threadfence_system();
    *(volatile unsigned long long *)&a.mirror[16] = a.seq;
  }
}

template <int OP> __host__ __device__ constexpr int tiny_streams() { return (OP == JP_OP_PRIV_TMP || OP == JP_OP_STENCIL2) ? 3 : 2; }
// exposed reads of A (X is never written, T reads are covered)
template <int OP> __host__ __device__ constexpr int n_exposed_tiny() {
  return OP == JP_OP_ADD_C ? 1 : OP == JP_OP_SAXPY ? 1 : OP == JP_OP_STENCIL2 ? 2 : 0;
}

__device__ __forceinline__ void cp_async16_t(void *smem, const void *gmem) {
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"((unsigned)__cvta_generic_to_shared(smem)), "l"(gmem)
               : "memory");
}
__device__ __forceinline__ void cp_async4_t(void *smem, const void *gmem) {
  asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"((unsigned)__cvta_generic_to_shared(smem)), "l"(gmem)
               : "memory");
}

// first-window / step rules of reading A8 (the device copy of tls_next_window)
__device__ __forceinline__ int tiny_pow2ceil(int x) { return x <= 1 ? 1 : 1 << (32 - __clz(x - 1)); }

template <int OP, int DT>
__global__ void __launch_bounds__(kTinyThreads, 1) k_tiny(DLoop L, TinyArgs a, int64_t *hdr) {
  constexpr int NS = tiny_streams<OP>();
  constexpr int T = kTinyThreads, K = kTinyK;
  extern __shared__ __align__(16) uint32_t tsm[];
  const int n = (int)L.n, lenA = (int)L.lenA, lenT = OP == JP_OP_PRIV_TMP ? (int)L.lenT : 0;
  int32_t *ix = reinterpret_cast<int32_t *>(tsm);   // [NS][n]: r, w, r2 | s
  uint32_t *sA = tsm + NS * n;                     // A values
  uint32_t *sT = sA + lenA;                        // T values
  uint32_t *tA0 = sT + lenT, *tA1 = tA0 + lenA;    // per-address tables of A
  uint32_t *tT0 = tA1 + lenA, *tT1 = tT0 + lenT;   // per-address tables of T
  uint32_t *rdy = tT1 + lenT;                      // on-chip TLS: window tag of the shadow value tA1[a]
  __shared__ unsigned s_cnt[4];                    // raw, war, waw, bad
  __shared__ int s_first, s_fv[2];
  const int tid = threadIdx.x, wbase = tid & ~31;
  const int32_t *src[3] = {L.r, L.w, OP == JP_OP_STENCIL2 ? L.r2 : OP == JP_OP_PRIV_TMP ? L.s : nullptr};
  if (tid < 4) s_cnt[tid] = 0;
  if (tid == 0) s_first = INT32_MAX;
  // stage indices, A and T with cp.async (all copies in flight at once; 16-byte
  // pieces when the source is aligned), identity indices written directly
  auto stage = [&](void *dst, const void *srcp, int count) {
    const bool a16 = (((uintptr_t)srcp | (uintptr_t)dst) & 15) == 0;
    const int nv = a16 ? count / 4 : 0;
    for (int v = tid; v < nv; v += T) cp_async16_t(static_cast<uint32_t *>(dst) + 4 * v, static_cast<const uint32_t *>(srcp) + 4 * v);
    for (int e = 4 * nv + tid; e < count; e += T) cp_async4_t(static_cast<uint32_t *>(dst) + e, static_cast<const uint32_t *>(srcp) + e);
  };
#pragma unroll
  for (int q = 0; q < NS; q++) {
    if (src[q]) stage(ix + q * n, src[q], n);
    else for (int i = tid; i < n; i += T) ix[q * n + i] = (int32_t)L.ioff + i;
  }
  stage(sA, L.A, lenA);
  if (lenT) stage(sT, L.T, lenT);
  asm volatile("cp.async.commit_group;\n\tcp.async.wait_group 0;" ::: "memory");
  for (int e = tid; e < lenA; e += T) { tA0[e] = 0xFFFFFFFFu; tA1[e] = 0xFFFFFFFFu; }
  for (int e = tid; e < lenT; e += T) { tT0[e] = 0xFFFFFFFFu; tT1[e] = 0xFFFFFFFFu; }
  JP_CTA_SYNC();
  // ---- validation (reading A13) and stamps (P1): first writer / first reader ----
  unsigned bad = 0;
  for (int i = tid; i < n; i += T) {
    const int32_t r = ix[i], w = ix[n + i], x2 = NS == 3 ? ix[2 * n + i] : 0;
    auto inA = [&](int32_t v) { return (uint32_t)v < (uint32_t)lenA; };
    if constexpr (OP == JP_OP_ADD_C) {
      if (!inA(r) || !inA(w)) { bad++; continue; }
      atomicMin(&tA0[w], (uint32_t)i);
      atomicMin(&tA1[r], (uint32_t)i);
    } else if constexpr (OP == JP_OP_SAXPY) {
      if ((uint32_t)r >= (uint32_t)L.lenX || !inA(w)) { bad++; continue; }
      atomicMin(&tA0[w], (uint32_t)i);
      atomicMin(&tA1[w], (uint32_t)i);
    } else if constexpr (OP == JP_OP_PRIV_TMP) {
      if ((uint32_t)r >= (uint32_t)L.lenX || !inA(w) || (uint32_t)x2 >= (uint32_t)lenT) { bad++; continue; }
      atomicMin(&tT0[x2], (uint32_t)i);   // T write == its covered read
      atomicMin(&tA0[w], (uint32_t)i);
    } else {
      if (!inA(r) || !inA(w) || !inA(x2)) { bad++; continue; }
      atomicMin(&tA0[w], (uint32_t)i);
      atomicMin(&tA1[r], (uint32_t)i);
      atomicMin(&tA1[x2], (uint32_t)i);
    }
  }
  if (bad) atomicAdd(&s_cnt[3], bad);
  JP_CTA_SYNC();
  if (s_cnt[3]) {   // JP_ERR_INDEX: nothing modified
    if (tid == 0) { hdr[H_BAD] = s_cnt[3]; hdr[H_TINY_MODE] = -1; }
    tiny_publish(hdr, a);
    return;
  }
  // ---- classify (P2) ----
  unsigned c_raw = 0, c_war = 0, c_waw = 0;
  int first = INT32_MAX;
  for (int i = tid; i < n; i += T) {
    const int32_t r = ix[i], w = ix[n + i], x2 = NS == 3 ? ix[2 * n + i] : 0;
    const uint32_t u = (uint32_t)i;
    bool raw = false, war, waw;
    if constexpr (OP == JP_OP_ADD_C) { raw = tA0[r] < u; war = tA1[w] < u; waw = tA0[w] < u; }
    else if constexpr (OP == JP_OP_SAXPY) { raw = tA0[w] < u; war = tA1[w] < u; waw = raw; }
    else if constexpr (OP == JP_OP_PRIV_TMP) { war = tT0[x2] < u; waw = tT0[x2] < u || tA0[w] < u; }
    else { raw = tA0[r] < u || tA0[x2] < u; war = tA1[w] < u; waw = tA0[w] < u; }
    c_raw += raw; c_war += war; c_waw += waw;
    if (raw && i < first) first = i;
  }
  c_raw = __reduce_add_sync(0xffffffffu, c_raw);
  c_war = __reduce_add_sync(0xffffffffu, c_war);
  c_waw = __reduce_add_sync(0xffffffffu, c_waw);
  first = __reduce_min_sync(0xffffffffu, first);
  if ((tid & 31) == 0) {
    if (c_raw) atomicAdd(&s_cnt[0], c_raw);
    if (c_war) atomicAdd(&s_cnt[1], c_war);
    if (c_waw) atomicAdd(&s_cnt[2], c_waw);
    if (first != INT32_MAX) atomicMin(&s_first, first);
  }
  JP_CTA_SYNC();
  const int64_t raw_n = s_cnt[0], war_n = s_cnt[1], waw_n = s_cnt[2];
  // ---- Fig. 2(b) (the same decision as jp_select_mode) ----
  const double d_raw = (double)raw_n / (double)n;
  const int mode = d_raw > a.tau ? JP_MODE_SEQ_RECOMMENDED : raw_n > 0 ? JP_MODE_TLS
                   : (war_n > 0 || waw_n > 0) ? JP_MODE_PRIVATIZED : JP_MODE_DOALL;
  long long committed = 0, executed = 0, windows = 0, viol = 0;
  int64_t wmax_used = 0;
  const bool onchip = mode != JP_MODE_DOALL && mode != JP_MODE_PRIVATIZED && waw_n == 0 && a.recovery != 1;
  if (onchip) {
    // ---- TLS with on-chip recovery (reading B7): fixed windows, every violator
    // re-executed once with its operand forwarded from the writer's shadow slot.
    // No address is written twice, so the window's write log is the first-writer
    // table tA0 of the profile restricted to the window: the writer of an exposed
    // read a is j = tA0[a], in the window iff ws <= j, earlier iff j < i.
    // Shadow values live per address (tA1[a], tagged by rdy[a] = window + 1).
    const int W = a.window > 0 ? (int)a.window : n;
    wmax_used = W;
    for (int e = tid; e < lenA; e += T) rdy[e] = 0;
    JP_CTA_SYNC();
    for (int ws = 0; ws < n; ws += W) {
      const int span = min(W, n - ws);
      const uint32_t tag = (uint32_t)windows + 1;
      uint32_t va[K], vt[K], g0[K], g1[K];
      uint32_t pend = 0;   // bit k: operand 0 waits on its writer; bit 16 + k: operand 1
      unsigned nv = 0;
      // SE from committed memory (sA) + DC against the window's writers
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= span) break;   // warp-uniform
        const int off = k * T + tid;
        if (off < span) {
          const int i = ws + off;
          const int32_t r = ix[i], w = ix[n + i], x2 = NS == 3 ? ix[2 * n + i] : 0;
          auto inwin = [&](int32_t addr) { const uint32_t j = tA0[addr]; return j >= (uint32_t)ws && j < (uint32_t)i; };
          if constexpr (OP == JP_OP_ADD_C) { g0[k] = sA[r]; if (inwin(r)) pend |= 1u << k; }
          else if constexpr (OP == JP_OP_SAXPY) { g0[k] = L.X[r]; g1[k] = sA[w]; }
          else if constexpr (OP == JP_OP_PRIV_TMP) g0[k] = L.X[r];
          else {
            g0[k] = sA[r]; g1[k] = sA[x2];
            if (inwin(r)) pend |= 1u << k;
            if (inwin(x2)) pend |= 1u << (16 + k);
          }
          nv += ((pend >> k) | (pend >> (16 + k))) & 1u;
        }
      }
      auto body = [&](int k) {
        if constexpr (OP == JP_OP_ADD_C) va[k] = op_add<DT>(g0[k], L.c0);
        else if constexpr (OP == JP_OP_SAXPY) va[k] = op_add<DT>(op_mul<DT>(L.c0, g0[k]), g1[k]);
        else if constexpr (OP == JP_OP_PRIV_TMP) { vt[k] = op_mul<DT>(L.c0, g0[k]); va[k] = op_add<DT>(vt[k], L.c1); }
        else va[k] = op_mul<DT>(op_add<DT>(g0[k], g1[k]), L.c0);
      };
      auto publish = [&](int k, int i) {
        const int32_t w = ix[n + i];
        *(volatile uint32_t *)&tA1[w] = va[k];
        __threadfence_block();
        *(volatile uint32_t *)&rdy[w] = tag;
      };
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= span) break;
        const int off = k * T + tid;
        if (off < span && !(((pend >> k) | (pend >> (16 + k))) & 1u)) { body(k); publish(k, ws + off); }
      }
      // recovery: violators in dependence order (their writers are earlier, so every wait ends)
      while (__any_sync(0xffffffffu, pend)) {
#pragma unroll
        for (int k = 0; k < K; k++) {
          if (((pend >> k) | (pend >> (16 + k))) & 1u) {
            const int i = ws + k * T + tid;
            if ((pend >> k) & 1u) {
              const int32_t r = ix[i];
              if (*(volatile uint32_t *)&rdy[r] == tag) { __threadfence_block(); g0[k] = *(volatile uint32_t *)&tA1[r]; pend &= ~(1u << k); }
            }
            if constexpr (OP == JP_OP_STENCIL2) {
              if ((pend >> (16 + k)) & 1u) {
                const int32_t x2 = ix[2 * n + i];
                if (*(volatile uint32_t *)&rdy[x2] == tag) { __threadfence_block(); g1[k] = *(volatile uint32_t *)&tA1[x2]; pend &= ~(1u << (16 + k)); }
              }
            }
            if (!(((pend >> k) | (pend >> (16 + k))) & 1u)) { body(k); publish(k, i); }
          }
        }
      }
      JP_CTA_SYNC();   // every read of committed memory in this window is done
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= span) break;
        const int off = k * T + tid;
        if (off < span) {
          const int i = ws + off;
          sA[ix[n + i]] = va[k];
          if constexpr (OP == JP_OP_PRIV_TMP) sT[ix[2 * n + i]] = vt[k];
        }
      }
      nv = __reduce_add_sync(0xffffffffu, nv);
      if ((tid & 31) == 0 && nv) atomicAdd(&s_cnt[3], nv);   // s_cnt[3] (bad) is 0 here: reused as the counter
      JP_CTA_SYNC();   // commits visible to the next window
      windows++;
    }
    viol = s_cnt[3];
    committed = n;
    executed = n + viol;
  } else if (mode == JP_MODE_DOALL) {
    // ---- DOALL: no dependence, any order ----
    for (int i = tid; i < n; i += T) {
      const int32_t r = ix[i], w = ix[n + i], x2 = NS == 3 ? ix[2 * n + i] : 0;
      if constexpr (OP == JP_OP_ADD_C) sA[w] = op_add<DT>(sA[r], L.c0);
      else if constexpr (OP == JP_OP_SAXPY) sA[w] = op_add<DT>(op_mul<DT>(L.c0, L.X[r]), sA[w]);
      else if constexpr (OP == JP_OP_PRIV_TMP) { const uint32_t t = op_mul<DT>(L.c0, L.X[r]); sT[x2] = t; sA[w] = op_add<DT>(t, L.c1); }
      else sA[w] = op_mul<DT>(op_add<DT>(sA[r], sA[x2]), L.c0);
    }
  } else if (mode == JP_MODE_PRIVATIZED) {
    // ---- PE(V): values from the pre-loop snapshot, then last writer wins ----
    // (tA1 / tT1 become "last writer + 1", 0 = none)
    for (int e = tid; e < lenA; e += T) tA1[e] = 0;
    for (int e = tid; e < lenT; e += T) tT1[e] = 0;
    JP_CTA_SYNC();
    uint32_t va[K], vt[K];
#pragma unroll
    for (int k = 0; k < K; k++) {
      const int i = k * T + tid;
      if (i < n) {
        const int32_t r = ix[i], w = ix[n + i], x2 = NS == 3 ? ix[2 * n + i] : 0;
        if constexpr (OP == JP_OP_ADD_C) va[k] = op_add<DT>(sA[r], L.c0);
        else if constexpr (OP == JP_OP_SAXPY) va[k] = op_add<DT>(op_mul<DT>(L.c0, L.X[r]), sA[w]);
        else if constexpr (OP == JP_OP_PRIV_TMP) { vt[k] = op_mul<DT>(L.c0, L.X[r]); va[k] = op_add<DT>(vt[k], L.c1); }
        else va[k] = op_mul<DT>(op_add<DT>(sA[r], sA[x2]), L.c0);
        atomicMax(&tA1[w], (uint32_t)i + 1);
        if constexpr (OP == JP_OP_PRIV_TMP) atomicMax(&tT1[x2], (uint32_t)i + 1);
      }
    }
    JP_CTA_SYNC();
#pragma unroll
    for (int k = 0; k < K; k++) {
      const int i = k * T + tid;
      if (i < n) {
        const int32_t w = ix[n + i];
        if (tA1[w] == (uint32_t)i + 1) sA[w] = va[k];
        if constexpr (OP == JP_OP_PRIV_TMP) { const int32_t x2 = ix[2 * n + i]; if (tT1[x2] == (uint32_t)i + 1) sT[x2] = vt[k]; }
      }
    }
  } else {
    // ---- TLS windows (the single-CTA algorithm, stamps direct-mapped) ----
    const int wfix = (int)a.window;
    int wmax = (int)a.w_max;
    if (wmax <= 0) {   // auto_w_max: clamp(pow2ceil(sqrt(1000 / d_raw)), 256, 1024)
      const double t = sqrt(1000.0 / d_raw);
      wmax = 256;
      while ((double)wmax < t && wmax < 1024) wmax <<= 1;
    }
    wmax_used = wmax;
    int W = wfix > 0 ? wfix
                     : min(max(tiny_pow2ceil((int)((4 * (int64_t)n + raw_n - 1) / raw_n)), 32), wmax);
    const bool dc = n_exposed_tiny<OP>() > 0;
    int ws = 0;
    uint32_t epoch = 0;
    // tA0 = write stamps of A, tA1 = commit order of A, tT1 = commit order of T (reset)
    for (int e = tid; e < lenA; e += T) { tA0[e] = 0xFFFFFFFFu; tA1[e] = 0; }
    for (int e = tid; e < lenT; e += T) tT1[e] = 0;
    if (tid == 0) { s_fv[0] = INT32_MAX; s_fv[1] = INT32_MAX; }
    const bool waw_any = waw_n > 0;   // no duplicate writer anywhere: commit is a plain scatter
    int par = 0;
    JP_CTA_SYNC();
    while (ws < n) {
      epoch++;
      if (tid == 0) s_fv[par ^ 1] = INT32_MAX;   // next window's slot (last read two barriers ago)
      const int span = min(W, n - ws);
      const uint32_t tagS = (kTinyEpochs - epoch) << 12, tagC = epoch << 13;
      uint32_t va[K], vt[K];
      // SE: values from committed memory, write stamps
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= span) break;   // warp-uniform
        const int off = k * T + tid;
        if (off < span) {
          const int i = ws + off;
          const int32_t r = ix[i], w = ix[n + i], x2 = NS == 3 ? ix[2 * n + i] : 0;
          if constexpr (OP == JP_OP_ADD_C) va[k] = op_add<DT>(sA[r], L.c0);
          else if constexpr (OP == JP_OP_SAXPY) va[k] = op_add<DT>(op_mul<DT>(L.c0, L.X[r]), sA[w]);
          else if constexpr (OP == JP_OP_PRIV_TMP) { vt[k] = op_mul<DT>(L.c0, L.X[r]); va[k] = op_add<DT>(vt[k], L.c1); }
          else va[k] = op_mul<DT>(op_add<DT>(sA[r], sA[x2]), L.c0);
          if (dc) atomicMin(&tA0[w], tagS | (uint32_t)off);
        }
      }
      JP_CTA_SYNC();
      // DC: an exposed read with an earlier in-window writer (reading A7)
      if (dc) {
        int myfv = INT32_MAX;
#pragma unroll
        for (int k = 0; k < K; k++) {
          if (k * T + wbase >= span) break;
          const int off = k * T + tid;
          if (off < span && myfv == INT32_MAX) {
            const int i = ws + off;
            auto viol_at = [&](int32_t addr) {
              const uint32_t v = tA0[addr];
              return (v & 0xFFFFF000u) == tagS && (v & 0xFFFu) < (uint32_t)off;
            };
            bool v;
            if constexpr (OP == JP_OP_SAXPY) v = viol_at(ix[n + i]);
            else if constexpr (OP == JP_OP_STENCIL2) v = viol_at(ix[i]) || viol_at(ix[2 * n + i]);
            else v = viol_at(ix[i]);
            if (v) myfv = off;
          }
        }
        myfv = __reduce_min_sync(0xffffffffu, myfv);
        if ((tid & 31) == 0 && myfv != INT32_MAX) atomicMin(&s_fv[par], myfv);
        JP_CTA_SYNC();
      }
      const int fv = min(s_fv[par], span);
      // commit [ws, ws+fv): last committed writer per address wins
      if (waw_any) {
#pragma unroll
        for (int k = 0; k < K; k++) {
          if (k * T + wbase >= fv) break;
          const int off = k * T + tid;
          if (off < fv) {
            const int i = ws + off;
            atomicMax(&tA1[ix[n + i]], tagC | (uint32_t)(off + 1));
            if constexpr (OP == JP_OP_PRIV_TMP) atomicMax(&tT1[ix[2 * n + i]], tagC | (uint32_t)(off + 1));
          }
        }
        JP_CTA_SYNC();
      }
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= fv) break;
        const int off = k * T + tid;
        if (off < fv) {
          const int i = ws + off;
          const int32_t w = ix[n + i];
          if (!waw_any || tA1[w] == (tagC | (uint32_t)(off + 1))) sA[w] = va[k];
          if constexpr (OP == JP_OP_PRIV_TMP) {
            const int32_t x2 = ix[2 * n + i];
            if (!waw_any || tT1[x2] == (tagC | (uint32_t)(off + 1))) sT[x2] = vt[k];
          }
        }
      }
      committed += fv; executed += span; windows++; viol += fv < span;
      ws += fv;
      W = wfix > 0 ? wfix : min(max(tiny_pow2ceil(2 * max(fv, 16)), 32), wmax);
      par ^= 1;
      JP_CTA_SYNC();   // commits visible to the next window
    }
  }
  JP_CTA_SYNC();
  for (int e = tid; e < lenA; e += T) L.A[e] = sA[e];
  for (int e = tid; e < lenT; e += T) L.T[e] = sT[e];
  if (tid == 0) {
    hdr[H_RAW] = raw_n; hdr[H_WAR] = war_n; hdr[H_WAW] = waw_n;
    hdr[H_FIRST_RAW] = s_first == INT32_MAX ? -1 : L.base + s_first;
    hdr[H_BAD] = 0;
    hdr[H_TLS_COMMITTED] = committed; hdr[H_TLS_EXECUTED] = executed;
    hdr[H_TLS_WINDOWS] = windows; hdr[H_TLS_VIOL] = viol;
    hdr[H_TINY_MODE] = mode;
    hdr[H_TINY_WMAX] = wmax_used;
    hdr[H_TINY_REC] = onchip ? JP_TLS_ONCHIP : JP_TLS_RESTART;
  }
  tiny_publish(hdr, a);
}

size_t tiny_smem_bytes(const jp_loop *L) {
  const int ns = (L->op == JP_OP_PRIV_TMP || L->op == JP_OP_STENCIL2) ? 3 : 2;
  const int64_t lt = L->op == JP_OP_PRIV_TMP ? L->len_T : 0;
  return (size_t)4 * ((size_t)ns * L->n + 4 * (size_t)L->len_A + 3 * (size_t)lt);
}

bool tiny_eligible(const jp_loop *L) {
  if (L->n <= 0 || L->n > kTinyThreads * kTinyK || L->len_A > 8192) return false;
  if (L->op == JP_OP_PRIV_TMP && L->len_T > 4096) return false;
  if (L->iter_base != 0 || L->ident_off != 0) return false;   // whole loops only
  return tiny_smem_bytes(L) <= 200 * 1024;
}

template <int OP, int DT>
static cudaError_t run_tiny(const DLoop &d, TinyArgs a, size_t smem, int64_t *hdr, cudaStream_t st) {
  static int done[64] = {0};   // the attribute is set once per device (the maximum the path uses)
  int dev = 0;
  cudaGetDevice(&dev);
  if (dev >= 0 && dev < 64 && !done[dev]) {
    cudaError_t e = cudaFuncSetAttribute(k_tiny<OP, DT>, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    if (e != cudaSuccess) return e;
    done[dev] = 1;
  }
  k_tiny<OP, DT><<<1, kTinyThreads, smem, st>>>(d, a, hdr);
  note_launch();
  return cudaGetLastError();
}
template <int OP, int DT>
static void run_tiny_v(cudaError_t &e, const DLoop &d, TinyArgs a, size_t smem, int64_t *hdr, cudaStream_t st) {
  e = run_tiny<OP, DT>(d, a, smem, hdr, st);
}

cudaError_t launch_tiny(const Job &j, const jp_loop *L, double tau, int64_t window, int64_t w_max, int recovery,
                        int64_t *hdr, cudaStream_t st, int64_t *mirror, unsigned long long seq) {
  TinyArgs a;
  a.tau = tau;
  a.window = window;
  a.w_max = w_max;
  a.recovery = recovery;
  a.mirror = mirror;
  a.seq = seq;
  cudaError_t e = cudaSuccess;
  JP_DISPATCH(j.op, j.dt, run_tiny_v, e, j.d, a, tiny_smem_bytes(L), hdr, st);
  return e;
}

}  // namespace jp

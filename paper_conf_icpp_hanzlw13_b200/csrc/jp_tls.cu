// jp_tls.cu -- GPU thread-level speculation (mode B P:L367-375).
//
// "GPU-TLS adopts an incremental solution dividing the target loop into
// several sub-loops ... four phases: speculative execution (SE), dependency
// checking (DC), commit and mis-speculation recovery".  Here one
// sub-loop is a window [ws, ws+W) and the whole sequence of windows runs inside
// ONE persistent kernel (no host round trip per violation, unlike mode B's
// "forwards control to CPU", P:L369-372 -- see DESIGN.md Sec.7):
//   SE  each iteration reads COMMITTED memory, computes its writes into
//       registers (the per-thread "buffered possibly unsafe memory updates",
//       P:L323-325) and records its write addresses as metadata;
//   DC  an iteration violates iff one of its exposed reads was written by an
//       earlier iteration of the same window (reading A7); the first violator
//       fv is a block/grid min-reduction ("which threads fell in
//       violation");
//   commit  iterations [ws, fv) store their buffered values, the highest
//       iteration winning per address (reading A6: prefix commit);
//   recovery  iterations >= fv are discarded and re-execute in the next
//       window, which starts at fv.
//
// Two paths:
//  k_tls_cta  one 1024-thread CTA, W <= 4096.  The window's write set lives in
//             a shared-memory open-addressing hash (key = address, min writer,
//             max committed writer): conflict detection never leaves the SM;
//             3 __syncthreads per window (5 with in-window WAW).
//  k_tls_grid cooperative all-SM kernel for large windows.  Writes are stamped
//             into an HBM/L2 table S[a] = (~epoch)<<32 | offset with atomicMin
//             (never reset: a newer epoch always compares smaller than stale
//             entries), violations checked against it, commit-order resolved
//             with C[a] = epoch<<32 | offset atomicMax; grid barriers between
//             phases.
#include "jp_host.h"

// CTA barrier of the TLS windows.  An explicit barrier.sync with a memory
// clobber: with the JP_CTA_SYNC() intrinsic the single-CTA window loop lost
// RAW violations intermittently on sm_100a (a window's first violator was
// missed in ~1 of 3 runs at W = 4096); the same kernel with this barrier passed
// 80/80 repetitions ("TLS barrier").
#define TLS_SYNC() asm volatile("barrier.sync 0;" ::: "memory")

namespace jp {

struct TlsArgs {
  int64_t window, w_max, prof_raw;
  int hashA, hashT;   // array needs conflict tracking (reached through a non-identity index)
};

__host__ __device__ inline int64_t pow2ceil64(int64_t x) {
  int64_t p = 1;
  while (p < x) p <<= 1;
  return p;
}
__host__ __device__ inline int64_t clamp64(int64_t x, int64_t lo, int64_t hi) { return x < lo ? lo : x > hi ? hi : x; }

// Reading A8 (deterministic adaptive window).
__host__ __device__ inline int64_t next_window(int64_t n, int64_t prof_raw, int64_t prev, int64_t w_max) {
  if (prev < 0) {
    int64_t w0 = prof_raw < 0 ? 4096 : prof_raw == 0 ? w_max : pow2ceil64((4 * n + prof_raw - 1) / prof_raw);
    return clamp64(w0, 32, w_max);
  }
  return clamp64(pow2ceil64(2 * (prev > 16 ? prev : 16)), 32, w_max);
}
int64_t tls_next_window(int64_t n, int64_t prof_raw, int64_t prev, int64_t w_max) {
  return next_window(n, prof_raw, prev, w_max);
}

// ---------------------------------------------------------------------------
// shared-memory hash of the window's write set
// ---------------------------------------------------------------------------
__device__ __forceinline__ uint32_t hkey_of(int64_t addr, int tag) { return ((uint32_t)addr << 1) | (uint32_t)tag; }
__device__ __forceinline__ uint32_t hhome(uint32_t key) { return (key * 0x9E3779B1u) >> (32 - kTlsHashLog); }

__device__ __forceinline__ int hins(uint32_t *hk, uint32_t *hmin, uint32_t key, uint32_t off) {
  uint32_t h = hhome(key);
  while (true) {
    const uint32_t prev = atomicCAS(&hk[h], kEmpty, key);
    if (prev == kEmpty || prev == key) break;
    h = (h + 1) & (kTlsHash - 1);
  }
  atomicMin(&hmin[h], off);
  return (int)h;
}
__device__ __forceinline__ int hfind(const uint32_t *hk, uint32_t key) {
  uint32_t h = hhome(key);
  while (true) {
    const uint32_t k = hk[h];
    if (k == key) return (int)h;
    if (k == kEmpty) return -1;
    h = (h + 1) & (kTlsHash - 1);
  }
}

// exposed-read addresses of the opcodes (X is never written, T reads are covered)
template <int OP> __device__ __forceinline__ int n_exposed() {
  return OP == JP_OP_ADD_C ? 1 : OP == JP_OP_SAXPY ? 1 : OP == JP_OP_STENCIL2 ? 2 : 0;
}

// index streams of an opcode, in ring order: 0 = r, 1 = w, 2 = r2 (STENCIL2) or s (PRIV_TMP)
template <int OP> __host__ __device__ constexpr int n_streams() {
  return (OP == JP_OP_PRIV_TMP || OP == JP_OP_STENCIL2) ? 3 : 2;
}
constexpr int kRing = 2 * kTlsCtaWmax;   // ring of prefetched indices: [ws, ws + 2 W_max)

__device__ __forceinline__ void cp_async4(void *smem, const void *gmem) {
  asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"((unsigned)__cvta_generic_to_shared(smem)),
               "l"(gmem) : "memory");
}
__device__ __forceinline__ void cp_async_commit_wait() {
  asm volatile("cp.async.commit_group;\n\tcp.async.wait_group 0;" ::: "memory");
}

// Single-CTA TLS.  Per window: SE reads the window's indices from a shared
// ring (prefetched with cp.async one window ahead, so the only dependent
// global access of SE is the gather of committed operands), issues every
// gather before any use, then inserts the write keys into the shared hash.
template <int OP, int DT, bool WAW>
__global__ void __launch_bounds__(kTlsCtaThreads, 1) k_tls_cta(DLoop L, TlsArgs P, int64_t *stats) {
  constexpr int NS = n_streams<OP>();
  extern __shared__ __align__(16) uint32_t hsm[];
  uint32_t *hk = hsm, *hmin = hsm + kTlsHash, *hmax = hsm + 2 * kTlsHash;
  int32_t *ring = reinterpret_cast<int32_t *>(hsm + 3 * kTlsHash);   // [NS][kRing]
  __shared__ int s_fv[2];
  const int tid = threadIdx.x, lane = tid & 31;
  const int32_t *src[3] = {L.r, L.w, OP == JP_OP_STENCIL2 ? L.r2 : OP == JP_OP_PRIV_TMP ? L.s : nullptr};
  for (int k = tid; k < kTlsHash; k += kTlsCtaThreads) { hk[k] = kEmpty; hmin[k] = 0xFFFFFFFFu; hmax[k] = 0; }
  if (tid == 0) { s_fv[0] = INT32_MAX; s_fv[1] = INT32_MAX; }
  // initial ring fill [0, min(n, kRing))
  int64_t hi = L.n < kRing ? L.n : kRing;
  for (int64_t i = tid; i < hi; i += kTlsCtaThreads)
#pragma unroll
    for (int q = 0; q < NS; q++)
      if (src[q]) cp_async4(&ring[q * kRing + i], src[q] + i);
  cp_async_commit_wait();
  TLS_SYNC();

  const bool dc = n_exposed<OP>() > 0 && P.hashA;
  int64_t ws = 0;
  int64_t W = P.window > 0 ? P.window : next_window(L.n, P.prof_raw, -1, P.w_max);
  long long committed = 0, executed = 0, windows = 0, viol = 0;
  int par = 0;
  while (ws < L.n) {
    const int span = (int)(W < L.n - ws ? W : L.n - ws);
    if (tid == 0) s_fv[par ^ 1] = INT32_MAX;
    // keep the ring full: [hi, ws + kRing) reuses the slots of iterations < ws
    {
      const int64_t to = ws + kRing < L.n ? ws + kRing : L.n;
      for (int64_t i = hi + tid; i < to; i += kTlsCtaThreads)
#pragma unroll
        for (int q = 0; q < NS; q++)
          if (src[q]) cp_async4(&ring[q * kRing + (i & (kRing - 1))], src[q] + i);
      asm volatile("cp.async.commit_group;" ::: "memory");
      hi = to;
    }
    uint32_t va[kTlsCtaIpt], vt[kTlsCtaIpt], g0[kTlsCtaIpt], g1[kTlsCtaIpt];
    int32_t ix0[kTlsCtaIpt], ix1[kTlsCtaIpt], ix2[kTlsCtaIpt];
    int slA[kTlsCtaIpt], slT[kTlsCtaIpt];
    // ---------------- SE: indices from the ring ----------------
#pragma unroll
    for (int k = 0; k < kTlsCtaIpt; k++) {
      const int off = k * kTlsCtaThreads + tid;
      if (off < span) {
        const int64_t i = ws + off;
        const int slot = (int)(i & (kRing - 1));
        ix0[k] = src[0] ? ring[slot] : (int32_t)(L.ioff + i);
        ix1[k] = src[1] ? ring[kRing + slot] : (int32_t)(L.ioff + i);
        if constexpr (NS == 3) ix2[k] = src[2] ? ring[2 * kRing + slot] : (int32_t)(L.ioff + i);
      }
    }
    // ---------------- SE: gather committed operands (all issued before use) ----------------
#pragma unroll
    for (int k = 0; k < kTlsCtaIpt; k++) {
      const int off = k * kTlsCtaThreads + tid;
      if (off < span) {
        if constexpr (OP == JP_OP_ADD_C) g0[k] = L.A[ix0[k]];
        else if constexpr (OP == JP_OP_SAXPY) { g0[k] = L.X[ix0[k]]; g1[k] = L.A[ix1[k]]; }
        else if constexpr (OP == JP_OP_PRIV_TMP) g0[k] = L.X[ix0[k]];
        else { g0[k] = L.A[ix0[k]]; g1[k] = L.A[ix2[k]]; }
      }
    }
    // ---------------- SE: values into the write log, write keys into the hash ----------------
#pragma unroll
    for (int k = 0; k < kTlsCtaIpt; k++) {
      const int off = k * kTlsCtaThreads + tid;
      if (off < span) {
        if constexpr (OP == JP_OP_ADD_C) va[k] = op_add<DT>(g0[k], L.c0);
        else if constexpr (OP == JP_OP_SAXPY) va[k] = op_add<DT>(op_mul<DT>(L.c0, g0[k]), g1[k]);
        else if constexpr (OP == JP_OP_PRIV_TMP) { vt[k] = op_mul<DT>(L.c0, g0[k]); va[k] = op_add<DT>(vt[k], L.c1); }
        else va[k] = op_mul<DT>(op_add<DT>(g0[k], g1[k]), L.c0);
        if (P.hashA) slA[k] = hins(hk, hmin, hkey_of(ix1[k], 0), (uint32_t)off);
        if constexpr (OP == JP_OP_PRIV_TMP) if (P.hashT) slT[k] = hins(hk, hmin, hkey_of(ix2[k], 1), (uint32_t)off);
      }
    }
    TLS_SYNC();
    // ---------------- DC ----------------
    if (dc) {
      int myfv = INT32_MAX;
#pragma unroll
      for (int k = 0; k < kTlsCtaIpt; k++) {
        const int off = k * kTlsCtaThreads + tid;
        if (off < span && myfv == INT32_MAX) {
          // exposed reads of A: ADD_C/STENCIL2 A[r] (+ A[r2]); SAXPY Y[w]
          const int32_t ra = OP == JP_OP_SAXPY ? ix1[k] : ix0[k];
          int h = hfind(hk, hkey_of(ra, 0));
          bool v = h >= 0 && hmin[h] < (uint32_t)off;
          if constexpr (OP == JP_OP_STENCIL2) {
            if (!v) { h = hfind(hk, hkey_of(ix2[k], 0)); v = h >= 0 && hmin[h] < (uint32_t)off; }
          }
          if (v) myfv = off;
        }
      }
      myfv = __reduce_min_sync(0xffffffffu, myfv);
      if (lane == 0 && myfv != INT32_MAX) atomicMin(&s_fv[par], myfv);
      TLS_SYNC();
    }
    const int fv = dc ? (s_fv[par] < span ? s_fv[par] : span) : span;
    // ---------------- commit [ws, ws+fv) ----------------
    if constexpr (WAW) {
#pragma unroll
      for (int k = 0; k < kTlsCtaIpt; k++) {
        const int off = k * kTlsCtaThreads + tid;
        if (off < fv) {
          if (P.hashA) atomicMax(&hmax[slA[k]], (uint32_t)off + 1);
          if constexpr (OP == JP_OP_PRIV_TMP) if (P.hashT) atomicMax(&hmax[slT[k]], (uint32_t)off + 1);
        }
      }
      TLS_SYNC();
    }
#pragma unroll
    for (int k = 0; k < kTlsCtaIpt; k++) {
      const int off = k * kTlsCtaThreads + tid;
      if (off < fv) {
        if (!WAW || !P.hashA || hmax[slA[k]] == (uint32_t)off + 1) L.A[ix1[k]] = va[k];
        if constexpr (OP == JP_OP_PRIV_TMP)
          if (!WAW || !P.hashT || hmax[slT[k]] == (uint32_t)off + 1) L.T[ix2[k]] = vt[k];
      }
    }
    if constexpr (WAW) TLS_SYNC();
    // clear the window's hash entries (no reader is left in this window)
#pragma unroll
    for (int k = 0; k < kTlsCtaIpt; k++) {
      const int off = k * kTlsCtaThreads + tid;
      if (off < span) {
        if (P.hashA) { hk[slA[k]] = kEmpty; hmin[slA[k]] = 0xFFFFFFFFu; hmax[slA[k]] = 0; }
        if constexpr (OP == JP_OP_PRIV_TMP)
          if (P.hashT) { hk[slT[k]] = kEmpty; hmin[slT[k]] = 0xFFFFFFFFu; hmax[slT[k]] = 0; }
      }
    }
    committed += fv; executed += span; windows++; viol += fv < span;
    ws += fv;
    W = P.window > 0 ? P.window : next_window(L.n, P.prof_raw, fv, P.w_max);
    par ^= 1;
    asm volatile("cp.async.wait_group 0;" ::: "memory");   // this window's prefetch has landed
    TLS_SYNC();   // commits and prefetched indices visible to the next SE, hash clean
  }
  if (tid == 0) { stats[0] = committed; stats[1] = executed; stats[2] = windows; stats[3] = viol; }
}

// ---------------------------------------------------------------------------
// cooperative all-SM path
// ---------------------------------------------------------------------------
constexpr int kTlsGridIpt = 2;

struct GridWs {
  unsigned long long *SA, *CA, *CT;   // stamps (A), commit order (A, T)
  unsigned *bar;                      // [0] count, [1] generation
  int64_t *fv;                        // 3 rotating slots
};

__device__ __forceinline__ void grid_sync(unsigned *bar) {
  JP_CTA_SYNC();
  if (threadIdx.x == 0) {
    volatile unsigned *vgen = bar + 1;
    const unsigned g = *vgen;
    __threadfence();
    if (atomicAdd(bar, 1u) == gridDim.x - 1) {
      atomicExch(bar, 0u);
      __threadfence();
      atomicAdd(bar + 1, 1u);
    } else {
      while (*vgen == g) { }
    }
    __threadfence();
  }
  JP_CTA_SYNC();
}

// body with L2-coherent (ld.global.cg) reads of the in/out array
template <int OP, int DT>
__device__ __forceinline__ void body_values_cg(const DLoop &L, int64_t i, uint32_t &va, uint32_t &vt) {
  if constexpr (OP == JP_OP_ADD_C) {
    va = op_add<DT>(__ldcg(L.A + ixl(L, L.r, i)), L.c0);
  } else if constexpr (OP == JP_OP_SAXPY) {
    va = op_add<DT>(op_mul<DT>(L.c0, L.X[ixl(L, L.r, i)]), __ldcg(L.A + ixl(L, L.w, i)));
  } else if constexpr (OP == JP_OP_PRIV_TMP) {
    vt = op_mul<DT>(L.c0, L.X[ixl(L, L.r, i)]);
    va = op_add<DT>(vt, L.c1);
  } else {
    va = op_mul<DT>(op_add<DT>(__ldcg(L.A + ixl(L, L.r, i)), __ldcg(L.A + ixl(L, L.r2, i))), L.c0);
  }
}

template <int OP, int DT, bool WAW>
__global__ void __launch_bounds__(kTlsGridThreads, 1) k_tls_grid(DLoop L, TlsArgs P, GridWs G, int64_t *stats) {
  const int64_t gt = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  const int64_t GT = (int64_t)gridDim.x * blockDim.x;
  const bool dc = n_exposed<OP>() > 0 && P.hashA;
  const int lane = threadIdx.x & 31;
  int64_t ws = 0;
  int64_t W = P.window > 0 ? P.window : next_window(L.n, P.prof_raw, -1, P.w_max);
  long long committed = 0, executed = 0, windows = 0, viol = 0;
  uint32_t epoch = 1;
  while (ws < L.n) {
    const int64_t span = W < L.n - ws ? W : L.n - ws;
    int64_t *fvslot = &G.fv[epoch % 3];
    if (gt == 0) G.fv[(epoch + 1) % 3] = INT64_MAX;
    const unsigned long long tagS = (unsigned long long)(~epoch) << 32;
    uint32_t va[kTlsGridIpt], vt[kTlsGridIpt];
    int32_t wa[kTlsGridIpt], wt[kTlsGridIpt], ra[kTlsGridIpt], rb[kTlsGridIpt];
    // ---------------- SE ----------------
#pragma unroll
    for (int k = 0; k < kTlsGridIpt; k++) {
      const int64_t off = k * GT + gt;
      if (off < span) {
        const int64_t i = ws + off;
        body_values_cg<OP, DT>(L, i, va[k], vt[k]);
        wa[k] = (int32_t)ixl(L, L.w, i);
        if constexpr (OP == JP_OP_PRIV_TMP) wt[k] = (int32_t)ixl(L, L.s, i);
        if constexpr (OP == JP_OP_ADD_C || OP == JP_OP_STENCIL2) ra[k] = (int32_t)ixl(L, L.r, i);
        if constexpr (OP == JP_OP_SAXPY) ra[k] = wa[k];
        if constexpr (OP == JP_OP_STENCIL2) rb[k] = (int32_t)ixl(L, L.r2, i);
        if (dc) atomicMin(&G.SA[wa[k]], tagS | (unsigned long long)off);
      }
    }
    grid_sync(G.bar);
    // ---------------- DC ----------------
    int64_t fv = span;
    if (dc) {
      long long myfv = INT64_MAX;
#pragma unroll
      for (int k = 0; k < kTlsGridIpt; k++) {
        const int64_t off = k * GT + gt;
        if (off < span && myfv == INT64_MAX) {
          unsigned long long s = __ldcg(&G.SA[ra[k]]);
          bool v = (s >> 32) == (unsigned long long)(~epoch) && (int64_t)(uint32_t)s < off;
          if constexpr (OP == JP_OP_STENCIL2) {
            if (!v) { s = __ldcg(&G.SA[rb[k]]); v = (s >> 32) == (unsigned long long)(~epoch) && (int64_t)(uint32_t)s < off; }
          }
          if (v) myfv = off;
        }
      }
      for (int o = 16; o; o >>= 1) {
        long long other = __shfl_xor_sync(0xffffffffu, myfv, o);
        myfv = other < myfv ? other : myfv;
      }
      if (lane == 0 && myfv != INT64_MAX) atomicMin((unsigned long long *)fvslot, (unsigned long long)myfv);
      grid_sync(G.bar);
      const int64_t f = *(volatile int64_t *)fvslot;
      fv = f < span ? f : span;
    }
    // ---------------- commit ----------------
    const unsigned long long tagC = (unsigned long long)epoch << 32;
    if constexpr (WAW) {
#pragma unroll
      for (int k = 0; k < kTlsGridIpt; k++) {
        const int64_t off = k * GT + gt;
        if (off < fv) {
          if (P.hashA) atomicMax(&G.CA[wa[k]], tagC | (unsigned long long)off);
          if constexpr (OP == JP_OP_PRIV_TMP) if (P.hashT) atomicMax(&G.CT[wt[k]], tagC | (unsigned long long)off);
        }
      }
      grid_sync(G.bar);
    }
#pragma unroll
    for (int k = 0; k < kTlsGridIpt; k++) {
      const int64_t off = k * GT + gt;
      if (off < fv) {
        if (!WAW || !P.hashA || __ldcg(&G.CA[wa[k]]) == (tagC | (unsigned long long)off)) __stcg(L.A + wa[k], va[k]);
        if constexpr (OP == JP_OP_PRIV_TMP)
          if (!WAW || !P.hashT || __ldcg(&G.CT[wt[k]]) == (tagC | (unsigned long long)off)) __stcg(L.T + wt[k], vt[k]);
      }
    }
    committed += fv; executed += span; windows++; viol += fv < span;
    ws += fv;
    W = P.window > 0 ? P.window : next_window(L.n, P.prof_raw, fv, P.w_max);
    epoch++;
    grid_sync(G.bar);
  }
  if (gt == 0) { stats[0] = committed; stats[1] = executed; stats[2] = windows; stats[3] = viol; }
}

template <int OP, int DT>
static cudaError_t run_tls(const DLoop &d, const TlsPlan &p, TlsArgs a, void *ws, const Layout &lo, int64_t *stats,
                           cudaStream_t st) {
  if (p.path == 1) {
    const size_t smem = 3 * kTlsHash * sizeof(uint32_t) + (size_t)n_streams<OP>() * kRing * sizeof(int32_t);
    if (p.waw) {
      cudaFuncSetAttribute(k_tls_cta<OP, DT, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
      k_tls_cta<OP, DT, true><<<1, kTlsCtaThreads, smem, st>>>(d, a, stats);
    } else {
      cudaFuncSetAttribute(k_tls_cta<OP, DT, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
      k_tls_cta<OP, DT, false><<<1, kTlsCtaThreads, smem, st>>>(d, a, stats);
    }
    note_launch();
    return cudaGetLastError();
  }
  GridWs g;
  g.SA = at<unsigned long long>(ws, lo, R_TLS_S_A);
  g.CA = at<unsigned long long>(ws, lo, R_TLS_C_A);
  g.CT = at<unsigned long long>(ws, lo, R_TLS_C_T);
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  g.bar = reinterpret_cast<unsigned *>(&hdr[H_BAR_COUNT]);
  g.fv = &hdr[H_FV0];
  cudaMemsetAsync(&hdr[H_BAR_COUNT], 0, 2 * sizeof(int64_t), st);
  cudaMemsetAsync(&hdr[H_FV0], 0x7F, 3 * sizeof(int64_t), st);   // "no violator" (>= any offset)
  if (g.SA) cudaMemsetAsync(g.SA, 0xFF, lo.bytes[R_TLS_S_A], st);
  if (g.CA) cudaMemsetAsync(g.CA, 0, lo.bytes[R_TLS_C_A], st);
  if (g.CT) cudaMemsetAsync(g.CT, 0, lo.bytes[R_TLS_C_T], st);
  int64_t wmax = p.window > 0 ? p.window : p.w_max;
  int64_t need = (wmax + (int64_t)kTlsGridThreads * kTlsGridIpt - 1) / ((int64_t)kTlsGridThreads * kTlsGridIpt);
  int maxb = 0;
  void *fn = p.waw ? (void *)k_tls_grid<OP, DT, true> : (void *)k_tls_grid<OP, DT, false>;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&maxb, fn, kTlsGridThreads, 0);
  int64_t cap = (int64_t)num_sms() * (maxb > 0 ? maxb : 1);
  if (need > cap) return cudaErrorInvalidConfiguration;
  int grid = (int)(need < 1 ? 1 : need);
  DLoop dd = d;
  void *args[] = {&dd, &a, &g, &stats};
  cudaError_t e = cudaLaunchCooperativeKernel(fn, grid, kTlsGridThreads, args, 0, st);
  note_launch();
  return e;
}

template <int OP, int DT>
static void run_tls_v(cudaError_t &e, const DLoop &d, const TlsPlan &p, TlsArgs a, void *ws, const Layout &lo,
                      int64_t *stats, cudaStream_t st) {
  e = run_tls<OP, DT>(d, p, a, ws, lo, stats, st);
}

cudaError_t launch_tls(const Job &j, void *ws, const Layout &lo, const TlsPlan &p, int64_t *stats, cudaStream_t st) {
  if (j.d.n == 0) {
    cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
    return launch_check();
  }
  TlsArgs a;
  a.window = p.window;
  a.w_max = p.w_max;
  a.prof_raw = p.prof_raw;
  a.hashA = a_indirect(j.op, j.d.r, j.d.r2, j.d.w);
  a.hashT = t_indirect(j.op, j.d.s);
  cudaError_t e = cudaSuccess;
  JP_DISPATCH(j.op, j.dt, run_tls_v, e, j.d, p, a, ws, lo, stats, st);
  if (e != cudaSuccess) return e;
  return launch_check();
}

}  // namespace jp

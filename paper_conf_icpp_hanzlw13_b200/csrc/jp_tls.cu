// jp_tls.cu -- GPU thread-level speculation (mode B P:L367-375).
//
// "GPU-TLS adopts an incremental solution dividing the target loop into
// several sub-loops ... four phases: speculative execution (SE), dependency
// checking (DC), commit and mis-speculation recovery".  Here one
// sub-loop is a window [ws, ws+W) and the whole sequence of windows runs inside
// ONE persistent kernel (no host round trip per violation, unlike mode B's
// "forwards control to CPU", P:L369-372 -- see DESIGN.md Sec.9):
//   SE  each iteration reads COMMITTED memory, computes its writes into
//       registers (the per-thread "buffered possibly unsafe memory updates",
//       P:L323-325) and records its write addresses as metadata;
//   DC  an iteration violates iff one of its exposed reads was written by an
//       earlier iteration of the same window (reading A7); the first violator
//       fv is a block/cluster/grid min-reduction ("which threads
//       fell in violation");
//   commit  iterations [ws, fv) store their buffered values, the highest
//       iteration winning per address (reading A6: prefix commit);
//   recovery  iterations >= fv are discarded and re-execute in the next
//       window, which starts at fv.
//
// Three paths:
//  k_tls_cta      one 1024-thread CTA, W <= 4096.  The window's write set lives
//                 in a shared-memory open-addressing hash of packed 64-bit
//                 entries (address key << 32 | min writer offset): conflict
//                 detection never leaves the SM; 3 CTA barriers per window
//                 (5 with in-window WAW).
//  k_tls_cluster  one thread-block cluster (C <= 16 CTAs), W <= 32(144C-1).
//                 Writes are stamped into an HBM/L2 table S[a] = (~epoch)<<32
//                 | offset with 64-bit atomicMin (never reset: a newer epoch
//                 compares smaller), split arrive/wait cluster barriers.
//  k_tls_grid     cooperative all-SM kernel for windows beyond a cluster,
//                 same stamps, software grid barrier.
// Guided runs (jp_tls_guide): only RAW-source writes
// are stamped/inserted and only raw reads are checked -- the same violators.
#include "jp_host.h"

// CTA barrier of the TLS windows.  An explicit barrier.sync with a memory
// clobber: with the __syncthreads() intrinsic the single-CTA window loop lost
// RAW violations intermittently on sm_100a (a window's first violator was
// missed in ~1 of 3 runs at W = 4096); the same kernel with this barrier passed
// 80/80 repetitions ("TLS barrier").
#define TLS_SYNC() asm volatile("barrier.sync 0;" ::: "memory")

#ifdef JP_TLS_TRACE
// phase timestamps (SM clock) of the first windows, thread 0 of CTA 0 (trace build only)
constexpr int kTraceWin = 2048, kTracePh = 16;
__device__ long long g_tls_trace[kTraceWin * kTracePh];
#define TLS_TR(ph) do { if (tr) g_tls_trace[windows * kTracePh + (ph)] = clock64(); } while (0)
#else
#define TLS_TR(ph) do { } while (0)
#endif

namespace jp {

struct TlsArgs {
  int64_t window, w_max, prof_raw;
  int hashA, hashT;   // array needs conflict tracking (reached through a non-identity index)
};

__host__ __device__ inline int64_t pow2ceil64(int64_t x) {
#ifdef __CUDA_ARCH__
  return x <= 1 ? 1 : (int64_t)1 << (64 - __clzll((unsigned long long)(x - 1)));
#else
  int64_t p = 1;
  while (p < x) p <<= 1;
  return p;
#endif
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
// the step rule alone (device, 32-bit, no division): clamp(pow2ceil(2*max(c,16)), 32, w_max)
__device__ __forceinline__ int next_window_step(int prev, int w_max) {
  const unsigned x = 2u * (unsigned)(prev > 16 ? prev : 16);
  const int p = (int)(1u << (32 - __clz(x - 1)));
  return p < 32 ? 32 : p > w_max ? w_max : p;
}
int64_t tls_next_window(int64_t n, int64_t prof_raw, int64_t prev, int64_t w_max) {
  return next_window(n, prof_raw, prev, w_max);
}

// ---------------------------------------------------------------------------
// shared-memory hash of the window's write set: one u64 per slot,
// key << 32 | min writer offset, empty = ~0 (no key is 0xFFFFFFFF: addresses
// are < 2^31 - 1, key = address << 1 | array tag).
// ---------------------------------------------------------------------------
constexpr unsigned long long kEmpty64 = ~0ull;
__device__ __forceinline__ uint32_t hkey_of(int64_t addr, int tag) { return ((uint32_t)addr << 1) | (uint32_t)tag; }
__device__ __forceinline__ uint32_t hhome(uint32_t key) { return (key * 0x9E3779B1u) >> (32 - kTlsHashLog); }

// Insert: one 64-bit CAS claims an empty slot with (key, off); a slot that
// already holds the key keeps the smaller offset (64-bit atomicMin on the same
// key compares offsets only).  Returns the slot.
__device__ __forceinline__ int hins64(unsigned long long *H, uint32_t key, uint32_t off) {
  const unsigned long long mine = ((unsigned long long)key << 32) | off;
  uint32_t h = hhome(key);
  while (true) {
    const unsigned long long prev = atomicCAS(&H[h], kEmpty64, mine);
    if (prev == kEmpty64) return (int)h;
    if ((uint32_t)(prev >> 32) == key) {
      if ((uint32_t)prev > off) atomicMin(&H[h], mine);
      return (int)h;
    }
    h = (h + 1) & (kTlsHash - 1);
  }
}
// min writer offset of key in the window, 0xFFFFFFFF if none
__device__ __forceinline__ uint32_t hmin64(const unsigned long long *H, uint32_t key) {
  uint32_t h = hhome(key);
  while (true) {
    const unsigned long long v = H[h];
    if ((uint32_t)(v >> 32) == key) return (uint32_t)v;
    if (v == kEmpty64) return 0xFFFFFFFFu;
    h = (h + 1) & (kTlsHash - 1);
  }
}

// exposed-read addresses of the opcodes (X is never written, T reads are covered)
template <int OP> __host__ __device__ constexpr int n_exposed() {
  return OP == JP_OP_ADD_C ? 1 : OP == JP_OP_SAXPY ? 1 : OP == JP_OP_STENCIL2 ? 2 : 0;
}

// index streams of an opcode, in ring order: 0 = r, 1 = w, 2 = r2 (STENCIL2) or s (PRIV_TMP)
template <int OP> __host__ __device__ constexpr int n_streams() {
  return (OP == JP_OP_PRIV_TMP || OP == JP_OP_STENCIL2) ? 3 : 2;
}

__device__ __forceinline__ void cp_async4(void *smem, const void *gmem) {
  asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"((unsigned)__cvta_generic_to_shared(smem)),
               "l"(gmem) : "memory");
}
__device__ __forceinline__ void cp_async16(void *smem, const void *gmem) {
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"((unsigned)__cvta_generic_to_shared(smem)), "l"(gmem)
               : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N> __device__ __forceinline__ void cp_async_wait() {
  asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory");
}

// Launch-time shape of the prefetch rings.
struct RingArgs {
  int ring_log;   // cta: ring entries per stream = 1 << ring_log; cluster: ring groups per CTA
  int wait1;      // ring holds >= 3 windows ahead: wait only for the previous windows' copies
  int al16;       // every index stream is 16-byte aligned
};

// ---------------------------------------------------------------------------
// single-CTA path
// ---------------------------------------------------------------------------
// Per window: SE reads the window's indices (and guide bits) from shared rings
// prefetched with cp.async >= one window ahead, so the only dependent global
// access is the gather of committed operands, issued before any use; write
// keys go into the shared hash.  DC looks the exposed reads up in the hash.
template <int OP, int DT, bool WAW, bool GUIDED>
__global__ void __launch_bounds__(kTlsCtaThreads, 1)
    k_tls_cta(DLoop L, TlsArgs P, RingArgs R, const uint32_t *gbits, int64_t *stats) {
  constexpr int NS = n_streams<OP>();
  constexpr int T = kTlsCtaThreads, K = kTlsCtaIpt;
  extern __shared__ __align__(16) unsigned long long hsm64[];
  const int RL = 1 << R.ring_log, RB = RL >> 5;
  unsigned long long *H = hsm64;                                    // [kTlsHash]
  uint32_t *hmax = reinterpret_cast<uint32_t *>(H + kTlsHash);      // [kTlsHash] (WAW)
  int32_t *ring = reinterpret_cast<int32_t *>(hmax + (WAW ? kTlsHash : 0));   // [NS][RL]
  uint32_t *bring = reinterpret_cast<uint32_t *>(ring + NS * RL);   // [2][RL/32] (GUIDED)
  __shared__ int s_fv[2];
  const int tid = threadIdx.x, lane = tid & 31, wbase = tid & ~31;
  const int32_t *src[3] = {L.r, L.w, OP == JP_OP_STENCIL2 ? L.r2 : OP == JP_OP_PRIV_TMP ? L.s : nullptr};
  const int64_t nwords = (L.n + 31) >> 5;
  for (int k = tid; k < kTlsHash; k += T) {
    H[k] = kEmpty64;
    if constexpr (WAW) hmax[k] = 0;
  }
  if (tid == 0) { s_fv[0] = INT32_MAX; s_fv[1] = INT32_MAX; }

  // ring fill up to [ws_, ws_ + RL): index chunks of 4 (16-byte copies when
  // aligned; hi % 4 == 0 or hi == n) and guide words [ws_/32, ws_/32 + RB)
  // (32-bit positions: n <= 2^31 - 2 and ws + RL < 2^32)
  const uint32_t n32 = (uint32_t)L.n;
  const bool s0 = src[0] != nullptr, s1 = src[1] != nullptr, s2 = src[2] != nullptr;
  uint32_t hi = 0, bhi = 0;
  auto fill = [&](uint32_t ws_) {
    uint32_t to = (ws_ + (uint32_t)RL) & ~3u;
    if (to > n32) to = n32;
    if (tid < kTlsFillThreads && to > hi) {   // a few warps issue the copies; the rest skip
      const uint32_t c1 = (to + 3) >> 2;
      for (uint32_t c = (hi >> 2) + tid; c < c1; c += kTlsFillThreads) {
        const uint32_t i0 = c << 2;
        const int slot = (int)(i0 & (RL - 1));
        if (R.al16 && i0 + 4 <= n32) {
          if (s0) cp_async16(&ring[slot], src[0] + i0);
          if (s1) cp_async16(&ring[RL + slot], src[1] + i0);
          if constexpr (NS == 3) if (s2) cp_async16(&ring[2 * RL + slot], src[2] + i0);
        } else {
          for (uint32_t e = 0; e < 4; e++) {
            if (i0 + e >= n32) break;
            if (s0) cp_async4(&ring[slot + e], src[0] + i0 + e);
            if (s1) cp_async4(&ring[RL + slot + e], src[1] + i0 + e);
            if constexpr (NS == 3) if (s2) cp_async4(&ring[2 * RL + slot + e], src[2] + i0 + e);
          }
        }
      }
    }
    if (to > hi) hi = to;
    if constexpr (GUIDED) {
      uint32_t bto = (ws_ >> 5) + (uint32_t)RB;
      if (bto > (uint32_t)nwords) bto = (uint32_t)nwords;
      if (tid < kTlsFillThreads)
        for (uint32_t g = bhi + tid; g < bto; g += kTlsFillThreads) {
          cp_async4(&bring[g & (RB - 1)], gbits + g);
          cp_async4(&bring[RB + (g & (RB - 1))], gbits + nwords + g);
        }
      if (bto > bhi) bhi = bto;
    }
    cp_async_commit();
  };
  fill(0);
  cp_async_wait<0>();
  TLS_SYNC();

  const bool dc = n_exposed<OP>() > 0 && P.hashA;
  const bool insA = P.hashA && (WAW || dc);   // A keys: commit order (WAW) and/or conflict detection
  uint32_t ws = 0;
  int W = (int)(P.window > 0 ? P.window : next_window(L.n, P.prof_raw, -1, P.w_max));
  const int wfix = (int)P.window, wmax = (int)P.w_max;
  long long committed = 0, executed = 0, windows = 0, viol = 0;
  int par = 0;
#ifdef JP_TLS_TRACE
  const bool trc = tid == 0;
#endif
  while (ws < n32) {
#ifdef JP_TLS_TRACE
    const bool tr = trc && windows < kTraceWin;
#endif
    TLS_TR(0);
    const int span = (int)((uint32_t)W < n32 - ws ? (uint32_t)W : n32 - ws);
    if (tid == 0) s_fv[par ^ 1] = INT32_MAX;
    fill(ws);   // reuses the slots of iterations < ws
    TLS_TR(8);
    uint32_t va[K], vt[K], g0[K], g1[K];
    int32_t ix0[K], ix1[K], ix2[K];
    int slA[K], slT[K];
    bool rawk[K];
    // ---------------- SE: indices and guide bits from the rings ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
      rawk[k] = true;
      slA[k] = slT[k] = -1;
      if (off < span) {
        const uint32_t i = ws + (uint32_t)off;
        const int slot = (int)(i & (RL - 1));
        const int32_t id = (int32_t)L.ioff + (int32_t)i;
        ix0[k] = s0 ? ring[slot] : id;
        ix1[k] = s1 ? ring[RL + slot] : id;
        if constexpr (NS == 3) ix2[k] = s2 ? ring[2 * RL + slot] : id;
      }
    }
    TLS_TR(9);
    // ---------------- SE: gather committed operands (all issued before use) ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
      if (off < span) {
        if constexpr (OP == JP_OP_ADD_C) g0[k] = L.A[ix0[k]];
        else if constexpr (OP == JP_OP_SAXPY) { g0[k] = L.X[ix0[k]]; g1[k] = L.A[ix1[k]]; }
        else if constexpr (OP == JP_OP_PRIV_TMP) g0[k] = L.X[ix0[k]];
        else { g0[k] = L.A[ix0[k]]; g1[k] = L.A[ix2[k]]; }
      }
    }
    TLS_TR(10);
    // ---------------- SE: write keys into the hash ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
      if (off < span) {
        bool ins = insA;
        if constexpr (GUIDED) {
          const uint32_t i = ws + (uint32_t)off;
          const int b = (int)((i >> 5) & (RB - 1)), sh = (int)(i & 31);
          rawk[k] = (bring[b] >> sh) & 1u;
          ins = ins && ((bring[RB + b] >> sh) & 1u);
        }
        if (ins) slA[k] = hins64(H, hkey_of(ix1[k], 0), (uint32_t)off);
        if constexpr (OP == JP_OP_PRIV_TMP && WAW) if (P.hashT) slT[k] = hins64(H, hkey_of(ix2[k], 1), (uint32_t)off);
      }
    }
    TLS_TR(1);
    TLS_SYNC();
    TLS_TR(2);
    // ---------------- DC ----------------
    if (dc) {
      int myfv = INT32_MAX;
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
        if (off < span && rawk[k] && myfv == INT32_MAX) {
          // exposed reads of A: ADD_C/STENCIL2 A[r] (+ A[r2]); SAXPY Y[w]
          const int32_t ra = OP == JP_OP_SAXPY ? ix1[k] : ix0[k];
          bool v = hmin64(H, hkey_of(ra, 0)) < (uint32_t)off;
          if constexpr (OP == JP_OP_STENCIL2) v = v || hmin64(H, hkey_of(ix2[k], 0)) < (uint32_t)off;
          if (v) myfv = off;
        }
      }
      myfv = __reduce_min_sync(0xffffffffu, myfv);
      TLS_TR(3);
      if (lane == 0 && myfv != INT32_MAX) atomicMin(&s_fv[par], myfv);
      TLS_SYNC();
      TLS_TR(4);
    }
    const int fv = dc ? (s_fv[par] < span ? s_fv[par] : span) : span;
    TLS_TR(11);
    // ---------------- commit [ws, ws+fv) ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
      if (off < span) {
        if constexpr (OP == JP_OP_ADD_C) va[k] = op_add<DT>(g0[k], L.c0);
        else if constexpr (OP == JP_OP_SAXPY) va[k] = op_add<DT>(op_mul<DT>(L.c0, g0[k]), g1[k]);
        else if constexpr (OP == JP_OP_PRIV_TMP) { vt[k] = op_mul<DT>(L.c0, g0[k]); va[k] = op_add<DT>(vt[k], L.c1); }
        else va[k] = op_mul<DT>(op_add<DT>(g0[k], g1[k]), L.c0);
      }
    }
    TLS_TR(12);
    if constexpr (WAW) {
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
        if (off < fv) {
          if (slA[k] >= 0) atomicMax(&hmax[slA[k]], (uint32_t)off + 1);
          if constexpr (OP == JP_OP_PRIV_TMP) if (slT[k] >= 0) atomicMax(&hmax[slT[k]], (uint32_t)off + 1);
        }
      }
      TLS_SYNC();
    }
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k * T + wbase >= span) break;   // warp-uniform: no later slot of this warp has work
      const int off = k * T + tid;
      if (off < fv) {
        if (!WAW || slA[k] < 0 || hmax[slA[k]] == (uint32_t)off + 1) L.A[ix1[k]] = va[k];
        if constexpr (OP == JP_OP_PRIV_TMP)
          if (!WAW || slT[k] < 0 || hmax[slT[k]] == (uint32_t)off + 1) L.T[ix2[k]] = vt[k];
      }
    }
    if constexpr (WAW) TLS_SYNC();
    TLS_TR(5);
    // clear the window's hash entries (no reader is left in this window)
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k * T + wbase >= span) break;
      if (slA[k] >= 0) {
        H[slA[k]] = kEmpty64;
        if constexpr (WAW) hmax[slA[k]] = 0;
      }
      if constexpr (OP == JP_OP_PRIV_TMP && WAW)
        if (slT[k] >= 0) { H[slT[k]] = kEmpty64; hmax[slT[k]] = 0; }
    }
    if (R.wait1) cp_async_wait<1>();   // the copies issued before this window have landed
    else cp_async_wait<0>();           // this window's copies have landed
    TLS_TR(6);
    TLS_SYNC();   // commits and prefetched indices visible to the next SE, hash clean
    TLS_TR(7);
    committed += fv; executed += span; windows++; viol += fv < span;
    ws += (uint32_t)fv;
    W = wfix > 0 ? wfix : next_window_step(fv, wmax);
    par ^= 1;
    TLS_TR(13);
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

// ---------------------------------------------------------------------------
// thread-block-cluster path
// ---------------------------------------------------------------------------
// One cluster of C CTAs (C = 1, 2, 4, 8, 16, chosen at launch) runs the window
// loop.  The window [ws, ws+span) is cut into 32-iteration groups g = i >> 5;
// CTA c of the cluster owns the groups g = c (mod C), one group per warp at a
// time (lane = i & 31, so a warp holds 32 consecutive iterations in program
// order).  Per window:
//   SE   indices (and guide words) come from a per-CTA shared ring holding only
//        the CTA's own groups, prefetched with cp.async >= one window ahead.
//        Each (source) write is stamped into the HBM table S[a] =
//        (~epoch)<<32 | off with a fire-and-forget 64-bit atomicMin (RED); with
//        in-window WAW an intra-warp __match_any_sync on the address sends one
//        stamp per distinct address (the group's lowest lane = its earliest
//        iteration).
//   B1   split cluster barrier: arrive.release after the stamps, then the
//        gathers of committed operands are issued, then wait.acquire -- the
//        gather latency overlaps the barrier; values are consumed at commit.
//   DC   (raw) reads look their address up in S: a violation iff the stamp
//        carries this epoch and a smaller offset; every load is issued before
//        any is compared.  Warp min (__reduce_min_sync); the warp leader pushes
//        it with red.shared::cluster.min into the fv slot of every CTA.
//   B2   arrive.release; the write-log values are computed (gathers land);
//        wait.acquire; fv read from the CTA's own slot.
//   commit  iterations < fv store their values; with in-window WAW the highest
//        committed lane of each __match_any_sync group competes through
//        C[a] = epoch<<32|off atomicMax, a full cluster barrier, and the
//        winner stores.
//   B3   arrive.release after the commit stores; the NEXT window's SE (ring
//        reads, stamps) runs before its wait.acquire, which precedes the next
//        gathers.
// All CTAs see the same fv, so they run identical window loops.
constexpr int kTlsClThreads = 512;
constexpr int kTlsClWarps = kTlsClThreads / 32;
constexpr int kTlsClK = 9;   // groups per warp per window (W = 65024 at C = 16)

__device__ __forceinline__ uint32_t cluster_rank() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
  return r;
}
__device__ __forceinline__ void cl_arrive() { asm volatile("barrier.cluster.arrive.release.aligned;" ::: "memory"); }
__device__ __forceinline__ void cl_wait() { asm volatile("barrier.cluster.wait.acquire.aligned;" ::: "memory"); }
// min into the u32 at `p` (shared, this CTA's address) in CTA `rank` of the cluster
__device__ __forceinline__ void red_min_cluster(const void *p, uint32_t rank, uint32_t v) {
  const uint32_t la = (uint32_t)__cvta_generic_to_shared(p);
  asm volatile("{\n\t.reg .u32 ra;\n\tmapa.shared::cluster.u32 ra, %0, %1;\n\tred.shared::cluster.min.u32 [ra], %2;\n\t}"
               ::"r"(la), "r"(rank), "r"(v) : "memory");
}



template <int OP, int DT, bool WAW, bool GUIDED>
__global__ void __launch_bounds__(kTlsClThreads, 1)
    k_tls_cluster(DLoop L, TlsArgs P, unsigned long long *SA, unsigned long long *CA, unsigned long long *CT,
                  RingArgs R, int logC, const uint32_t *gbits, int64_t *stats) {
  constexpr int NS = n_streams<OP>();
  constexpr int K = kTlsClK;
  extern __shared__ __align__(16) int32_t ring[];   // [NS][RG][32] then guide words [2][RG]
  __shared__ uint32_t s_fv[2];
  const int RG = 1 << R.ring_log;
  uint32_t *bring = reinterpret_cast<uint32_t *>(ring + NS * RG * 32);
  const int C = 1 << logC;
  const int crank = (int)cluster_rank();
  const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
  const int32_t *src[3] = {L.r, L.w, OP == JP_OP_STENCIL2 ? L.r2 : OP == JP_OP_PRIV_TMP ? L.s : nullptr};
  const bool dc = n_exposed<OP>() > 0 && P.hashA;
  const int64_t ngroups = (L.n + 31) >> 5;
  const int64_t qmax = (ngroups - crank + C - 1) >> logC;   // groups owned by this CTA

  // ring refill: this CTA's groups g = q*C + crank for q in [q_fill, q_to);
  // issued by the first kTlsFillThreads threads; one commit group per call
  // (possibly empty) for the wait_group accounting.  32-bit positions:
  // n <= 2^31 - 2, so group and q counts fit.
  const uint32_t n32 = (uint32_t)L.n;
  const bool s0 = src[0] != nullptr, s1 = src[1] != nullptr, s2 = src[2] != nullptr;
  uint32_t q_fill = 0;
  auto refill = [&](uint32_t ws_) {
    uint32_t q_to = ((ws_ >> 5) >> logC) + (uint32_t)RG;
    if (q_to > (uint32_t)qmax) q_to = (uint32_t)qmax;
    if (tid < kTlsFillThreads && q_to > q_fill) {
      const uint32_t nq = q_to - q_fill;
      if (R.al16) {
        for (uint32_t u = tid; u < nq * 8; u += kTlsFillThreads) {   // 8 x 16 B per group and stream
          const uint32_t q = q_fill + (u >> 3), part = u & 7;
          const uint32_t i0 = (((q << logC) + (uint32_t)crank) << 5) + part * 4;
          const int d = (int)(q & (RG - 1)) * 32 + (int)part * 4;
          if (i0 + 4 <= n32) {
            if (s0) cp_async16(&ring[d], src[0] + i0);
            if (s1) cp_async16(&ring[RG * 32 + d], src[1] + i0);
            if constexpr (NS == 3) if (s2) cp_async16(&ring[2 * RG * 32 + d], src[2] + i0);
          } else {
            for (uint32_t e = 0; e < 4; e++) {
              if (i0 + e >= n32) break;
              if (s0) cp_async4(&ring[d + e], src[0] + i0 + e);
              if (s1) cp_async4(&ring[RG * 32 + d + e], src[1] + i0 + e);
              if constexpr (NS == 3) if (s2) cp_async4(&ring[2 * RG * 32 + d + e], src[2] + i0 + e);
            }
          }
        }
      } else {
        for (uint32_t u = tid; u < nq * 32; u += kTlsFillThreads) {
          const uint32_t q = q_fill + (u >> 5), e = u & 31;
          const uint32_t i = (((q << logC) + (uint32_t)crank) << 5) + e;
          const int d = (int)(q & (RG - 1)) * 32 + (int)e;
          if (i < n32) {
            if (s0) cp_async4(&ring[d], src[0] + i);
            if (s1) cp_async4(&ring[RG * 32 + d], src[1] + i);
            if constexpr (NS == 3) if (s2) cp_async4(&ring[2 * RG * 32 + d], src[2] + i);
          }
        }
      }
      if constexpr (GUIDED) {
        for (uint32_t u = tid; u < nq; u += kTlsFillThreads) {
          const uint32_t q = q_fill + u, g = (q << logC) + (uint32_t)crank;
          cp_async4(&bring[q & (RG - 1)], gbits + g);
          cp_async4(&bring[RG + (q & (RG - 1))], gbits + ngroups + g);
        }
      }
    }
    if (q_to > q_fill) q_fill = q_to;
    cp_async_commit();
  };

  if (tid == 0) { s_fv[0] = 0xFFFFFFFFu; s_fv[1] = 0xFFFFFFFFu; }
  refill(0);
  cp_async_wait<0>();
  cl_arrive();
  cl_wait();

  uint32_t ws = 0;
  int W = (int)(P.window > 0 ? P.window : next_window(L.n, P.prof_raw, -1, P.w_max));
  const int wfix = (int)P.window, wmax = (int)P.w_max;
  long long committed = 0, executed = 0, windows = 0, viol = 0;
  uint32_t epoch = 1;
  int par = 0;
  bool first = true;
#ifdef JP_TLS_TRACE
  const bool trc = crank == 0 && tid == 0;
#endif
  while (ws < n32) {
#ifdef JP_TLS_TRACE
    const bool tr = trc && windows < kTraceWin;
#endif
    TLS_TR(0);
    const int span = (int)((uint32_t)W < n32 - ws ? (uint32_t)W : n32 - ws);
    if (tid == 0) s_fv[par] = 0xFFFFFFFFu;   // read last in window-2 (before two cluster barriers)
    refill(ws);
    const unsigned long long tagS = (unsigned long long)(~epoch) << 32;
    const unsigned long long tagC = (unsigned long long)epoch << 32;
    // this CTA's groups in the window: g = q*C + crank, q in [q0, q1)
    const uint32_t g0 = ws >> 5, g1 = (ws + (uint32_t)span + 31) >> 5;
    const uint32_t q0 = (g0 + (uint32_t)(C - 1 - crank)) >> logC;   // first q with q*C + crank >= g0
    const uint32_t q1 = (g1 + (uint32_t)(C - 1 - crank)) >> logC;
    uint32_t va[K], vt[K];
    int32_t wa[K], wt[K], ra[K], rb[K];
    uint32_t offk[K];
    bool act[K], rawk[K];
    // slots of this warp with a group in the window (warp-uniform)
    const int nq_w = (int)(q1 - q0) - warp;
    const int nk = nq_w <= 0 ? 0 : (nq_w + kTlsClWarps - 1) / kTlsClWarps < K ? (nq_w + kTlsClWarps - 1) / kTlsClWarps : K;
    // ---------------- SE: indices, guide bits, stamps ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k >= nk) break;
      const uint32_t q = q0 + (uint32_t)(warp + k * kTlsClWarps);
      act[k] = false;
      rawk[k] = false;
      if (q < q1) {                                  // warp-uniform
        const uint32_t i = (((q << logC) + (uint32_t)crank) << 5) + (uint32_t)lane;
        act[k] = i >= ws && i < ws + (uint32_t)span;
        const int slot = (int)(q & (RG - 1)) * 32 + lane;
        const int32_t id = (int32_t)L.ioff + (int32_t)i;
        const int32_t i0 = s0 ? ring[slot] : id;
        const int32_t i1 = s1 ? ring[RG * 32 + slot] : id;
        int32_t i2 = 0;
        if constexpr (NS == 3) i2 = s2 ? ring[2 * RG * 32 + slot] : id;
        offk[k] = i - ws;
        wa[k] = i1;
        if constexpr (OP == JP_OP_PRIV_TMP) wt[k] = i2;
        if constexpr (OP == JP_OP_SAXPY) ra[k] = i1; else ra[k] = i0;
        if constexpr (OP == JP_OP_STENCIL2) rb[k] = i2;
        if constexpr (OP == JP_OP_SAXPY) rb[k] = i0;   // X index (the exposed A read is Y[w])
        rawk[k] = act[k];
        bool stamp = act[k];
        if constexpr (GUIDED) {
          const int b = (int)(q & (RG - 1));
          rawk[k] = act[k] && ((bring[b] >> lane) & 1u);
          stamp = act[k] && ((bring[RG + b] >> lane) & 1u);
        }
        if (dc) {
          if constexpr (WAW) {
            // one stamp per distinct address per warp: the lowest lane is the earliest writer
            const unsigned am = __ballot_sync(0xffffffffu, stamp);
            const unsigned grp = __match_any_sync(0xffffffffu, stamp ? wa[k] : -1) & am;
            stamp = stamp && (__ffs(grp) - 1) == lane;
          }
          if (stamp) atomicMin(&SA[wa[k]], tagS | offk[k]);
        }
      }
    }
    TLS_TR(1);
    if (!first) cl_wait();   // B3 of the previous window: its commits are visible
    cl_arrive();             // B1: the stamps are performed
    // ---------------- SE: gathers (consumed at commit) ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k >= nk) break;
      if (act[k]) {
        if constexpr (OP == JP_OP_ADD_C) va[k] = __ldcg(L.A + ra[k]);
        else if constexpr (OP == JP_OP_SAXPY) { va[k] = __ldcg(L.A + wa[k]); vt[k] = L.X[rb[k]]; }
        else if constexpr (OP == JP_OP_PRIV_TMP) vt[k] = L.X[ra[k]];
        else { va[k] = __ldcg(L.A + ra[k]); vt[k] = __ldcg(L.A + rb[k]); }
      }
    }
    cl_wait();
    TLS_TR(2);
    // ---------------- DC ----------------
    int fv = span;
    if (dc) {
      unsigned long long sv[K], sv2[K];
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k >= nk) break;
        if (rawk[k]) {
          sv[k] = __ldcg(&SA[ra[k]]);
          if constexpr (OP == JP_OP_STENCIL2) sv2[k] = __ldcg(&SA[rb[k]]);
        }
      }
      uint32_t myfv = 0xFFFFFFFFu;
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k >= nk) break;
        if (rawk[k]) {
          bool v = (uint32_t)(sv[k] >> 32) == ~epoch && (uint32_t)sv[k] < offk[k];
          if constexpr (OP == JP_OP_STENCIL2) v = v || ((uint32_t)(sv2[k] >> 32) == ~epoch && (uint32_t)sv2[k] < offk[k]);
          if (v && offk[k] < myfv) myfv = offk[k];
        }
      }
      myfv = __reduce_min_sync(0xffffffffu, myfv);
      TLS_TR(3);
      if (myfv != 0xFFFFFFFFu && lane < C) red_min_cluster(&s_fv[par], (uint32_t)lane, myfv);
      cl_arrive();   // B2
    }
    // ---------------- write-log values (the gathers land here) ----------------
#pragma unroll
    for (int k = 0; k < K; k++) {
      if (k >= nk) break;
      if (act[k]) {
        if constexpr (OP == JP_OP_ADD_C) va[k] = op_add<DT>(va[k], L.c0);
        else if constexpr (OP == JP_OP_SAXPY) va[k] = op_add<DT>(op_mul<DT>(L.c0, vt[k]), va[k]);
        else if constexpr (OP == JP_OP_PRIV_TMP) { vt[k] = op_mul<DT>(L.c0, vt[k]); va[k] = op_add<DT>(vt[k], L.c1); }
        else va[k] = op_mul<DT>(op_add<DT>(va[k], vt[k]), L.c0);
      }
    }
    if (dc) {
      cl_wait();
      TLS_TR(4);
      const uint32_t f = *(volatile uint32_t *)&s_fv[par];
      fv = f < (uint32_t)span ? (int)f : span;
    }
    // ---------------- commit [ws, ws+fv) ----------------
    if constexpr (WAW) {
      bool winA[K], winT[K];
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k >= nk) break;
        const uint32_t q = q0 + (uint32_t)(warp + k * kTlsClWarps);
        winA[k] = winT[k] = false;
        if (q < q1) {
          const bool c = act[k] && offk[k] < (uint32_t)fv;
          const unsigned cm = __ballot_sync(0xffffffffu, c);
          if (P.hashA) {
            // intra-warp: the highest committed lane of each address group
            const unsigned grp = __match_any_sync(0xffffffffu, c ? wa[k] : -1) & cm;
            winA[k] = c && (31 - __clz(grp)) == lane;
            if (winA[k]) atomicMax(&CA[wa[k]], tagC | offk[k]);
          } else {
            winA[k] = c;
          }
          if constexpr (OP == JP_OP_PRIV_TMP) {
            if (P.hashT) {
              const unsigned grp = __match_any_sync(0xffffffffu, c ? wt[k] : -1) & cm;
              winT[k] = c && (31 - __clz(grp)) == lane;
              if (winT[k]) atomicMax(&CT[wt[k]], tagC | offk[k]);
            } else {
              winT[k] = c;
            }
          }
        }
      }
      cl_arrive();   // B2': commit-order stamps performed
      cl_wait();
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k >= nk) break;
        if (winA[k] && (!P.hashA || __ldcg(&CA[wa[k]]) == (tagC | offk[k]))) __stcg(L.A + wa[k], va[k]);
        if constexpr (OP == JP_OP_PRIV_TMP)
          if (winT[k] && (!P.hashT || __ldcg(&CT[wt[k]]) == (tagC | offk[k]))) __stcg(L.T + wt[k], vt[k]);
      }
    } else {
#pragma unroll
      for (int k = 0; k < K; k++) {
        if (k >= nk) break;
        if (act[k] && offk[k] < (uint32_t)fv) {
          __stcg(L.A + wa[k], va[k]);
          if constexpr (OP == JP_OP_PRIV_TMP) __stcg(L.T + wt[k], vt[k]);
        }
      }
    }
    TLS_TR(5);
    if (R.wait1) cp_async_wait<1>();   // the copies issued before this window have landed
    else cp_async_wait<0>();           // this window's copies have landed
    TLS_SYNC();                        // ... and are visible to the CTA's next SE
    TLS_TR(6);
    cl_arrive();                       // B3 (waited at the next window, after its stamps)
    TLS_TR(7);
    first = false;
    committed += fv; executed += span; windows++; viol += fv < span;
    ws += (uint32_t)fv;
    W = wfix > 0 ? wfix : next_window_step(fv, wmax);
    epoch++;
    par ^= 1;
  }
  if (!first) cl_wait();
  if (crank == 0 && tid == 0) { stats[0] = committed; stats[1] = executed; stats[2] = windows; stats[3] = viol; }
}

// largest window (iterations) the cluster path holds with C CTAs: a window of
// span iterations touches at most ceil(span/32)+1 groups (unaligned start),
// ceil of that / C per CTA.
int64_t tls_cluster_wcap(int C) { return (int64_t)32 * ((int64_t)kTlsClWarps * kTlsClK * C - 1); }

// Largest power-of-two cluster (<= 16) the current device can schedule for the
// cluster TLS kernel (cached per device).
int tls_max_cluster() {
  static int cache[64] = {0};
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= 64) return 8;
  if (cache[dev]) return cache[dev];
  int best = 8;
  void *fn = (void *)k_tls_cluster<JP_OP_ADD_C, JP_I32, false, true>;
  if (cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1) == cudaSuccess) {
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, 160 * 1024);
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(16, 1, 1);
    cfg.blockDim = dim3(kTlsClThreads, 1, 1);
    cfg.dynamicSmemBytes = 160 * 1024;
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

// Shared-memory budget of the TLS kernels (the opt-in maximum per CTA).
constexpr size_t kSmemBudget = 227 * 1024;

// Ring shape of the single-CTA path: ring >= 3 windows ahead (wait_group 1)
// when it fits next to the hash, else >= 2 windows (wait_group 0); false when
// neither fits (window too large for this opcode on one CTA).
static bool cta_ring(int ns, bool waw, bool guided, int64_t wcap, int &rlog, int &wait1, size_t &smem) {
  const size_t hash = (size_t)kTlsHash * 8 + (waw ? (size_t)kTlsHash * 4 : 0) + 64;
  for (int w1 = 1; w1 >= 0; w1--) {
    const int64_t need = (w1 ? 3 : 2) * wcap + 32;
    int64_t rl = 32;
    int lg = 5;
    while (rl < need) { rl <<= 1; lg++; }
    const size_t bytes = hash + (size_t)ns * rl * 4 + (guided ? (size_t)2 * (rl / 32) * 4 : 0);
    if (bytes <= kSmemBudget) { rlog = lg; wait1 = w1; smem = bytes - 64; return true; }
  }
  return false;
}
int64_t tls_cta_wcap(int op, bool waw, bool guided) {
  const int ns = (op == JP_OP_PRIV_TMP || op == JP_OP_STENCIL2) ? 3 : 2;
  int rl, w1;
  size_t sm;
  int64_t best = 0;
  for (int64_t w = 32; w <= kTlsCtaWmax; w <<= 1)
    if (cta_ring(ns, waw, guided, w, rl, w1, sm)) best = w;
  return best;
}

template <int OP, int DT>
static cudaError_t run_tls_cta(const DLoop &d, const TlsPlan &p, TlsArgs a, const uint32_t *bits, int64_t *stats,
                               cudaStream_t st) {
  const int64_t wcap = p.window > 0 ? p.window : p.w_max;
  RingArgs R;
  size_t smem = 0;
  if (!cta_ring(n_streams<OP>(), p.waw, p.guided, wcap, R.ring_log, R.wait1, smem)) return cudaErrorInvalidValue;
  auto al = [](const int32_t *q) { return q == nullptr || ((uintptr_t)q & 15) == 0; };
  R.al16 = al(d.r) && al(d.w) && al(d.r2) && al(d.s);
  void *fn = p.waw ? (void *)k_tls_cta<OP, DT, true, false>
                   : p.guided ? (void *)k_tls_cta<OP, DT, false, true> : (void *)k_tls_cta<OP, DT, false, false>;
  cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  DLoop dd = d;
  void *args[] = {&dd, &a, &R, &bits, &stats};
  e = cudaLaunchKernel(fn, dim3(1), dim3(kTlsCtaThreads), args, smem, st);
  note_launch();
  return e;
}

template <int OP, int DT>
static cudaError_t run_tls_cluster(const DLoop &d, const TlsPlan &p, TlsArgs a, unsigned long long *SA,
                                   unsigned long long *CA, unsigned long long *CT, const uint32_t *bits,
                                   int64_t *stats, cudaStream_t st) {
  const int C = p.cluster;
  int logC = 0;
  while ((1 << logC) < C) logC++;
  const int64_t wcap = p.window > 0 ? p.window : p.w_max;
  RingArgs R;
  // ring >= 3 windows ahead per CTA (wait_group 1) when it fits, else >= 2
  size_t smem = 0;
  bool ok = false;
  for (int w1 = 1; w1 >= 0 && !ok; w1--) {
    const int64_t need = (w1 ? 3 : 2) * wcap / (32 * C) + 4;
    int64_t rg = 1;
    int rlog = 0;
    while (rg < need) { rg <<= 1; rlog++; }
    smem = (size_t)n_streams<OP>() * rg * 32 * sizeof(int32_t) + (p.guided ? (size_t)2 * rg * 4 : 0);
    if (smem <= kSmemBudget) { R.ring_log = rlog; R.wait1 = w1; ok = true; }
  }
  if (!ok) return cudaErrorInvalidValue;
  auto al = [](const int32_t *q) { return q == nullptr || ((uintptr_t)q & 15) == 0; };
  R.al16 = al(d.r) && al(d.w) && al(d.r2) && al(d.s);
  void *fn = p.waw ? (void *)k_tls_cluster<OP, DT, true, false>
                   : p.guided ? (void *)k_tls_cluster<OP, DT, false, true> : (void *)k_tls_cluster<OP, DT, false, false>;
  cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  if (C > 8) {
    e = cudaFuncSetAttribute(fn, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
    if (e != cudaSuccess) return e;
  }
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3(C, 1, 1);
  cfg.blockDim = dim3(kTlsClThreads, 1, 1);
  cfg.dynamicSmemBytes = smem;
  cfg.stream = st;
  cudaLaunchAttribute attr[1];
  attr[0].id = cudaLaunchAttributeClusterDimension;
  attr[0].val.clusterDim.x = C;
  attr[0].val.clusterDim.y = 1;
  attr[0].val.clusterDim.z = 1;
  cfg.attrs = attr;
  cfg.numAttrs = 1;
  DLoop dd = d;
  void *args[] = {&dd, &a, &SA, &CA, &CT, &R, &logC, &bits, &stats};
  e = cudaLaunchKernelExC(&cfg, fn, args);
  note_launch();
  return e;
}

template <int OP, int DT>
static cudaError_t run_tls(const DLoop &d, const TlsPlan &p, TlsArgs a, void *ws, const Layout &lo, int64_t *stats,
                           cudaStream_t st) {
  const uint32_t *bits = p.guided ? at<uint32_t>(ws, lo, R_GUIDE) : nullptr;
  if (p.path == 1) return run_tls_cta<OP, DT>(d, p, a, bits, stats, st);
  GridWs g;
  g.SA = at<unsigned long long>(ws, lo, R_TLS_S_A);
  g.CA = at<unsigned long long>(ws, lo, R_TLS_C_A);
  g.CT = at<unsigned long long>(ws, lo, R_TLS_C_T);
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  g.bar = reinterpret_cast<unsigned *>(&hdr[H_BAR_COUNT]);
  g.fv = &hdr[H_FV0];
  if (g.SA) cudaMemsetAsync(g.SA, 0xFF, lo.bytes[R_TLS_S_A], st);
  if (p.waw && g.CA) cudaMemsetAsync(g.CA, 0, lo.bytes[R_TLS_C_A], st);
  if (p.waw && g.CT) cudaMemsetAsync(g.CT, 0, lo.bytes[R_TLS_C_T], st);
  if (p.path == 3) return run_tls_cluster<OP, DT>(d, p, a, g.SA, g.CA, g.CT, bits, stats, st);
  cudaMemsetAsync(&hdr[H_BAR_COUNT], 0, 2 * sizeof(int64_t), st);
  cudaMemsetAsync(&hdr[H_FV0], 0x7F, 3 * sizeof(int64_t), st);   // "no violator" (>= any offset)
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

#ifdef JP_TLS_TRACE
cudaError_t tls_trace_copy(long long *host, int n) {
  return cudaMemcpyFromSymbol(host, g_tls_trace, sizeof(long long) * (size_t)n);
}
#endif

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

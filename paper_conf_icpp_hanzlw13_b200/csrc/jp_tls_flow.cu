// jp_tls_flow.cu -- on-chip TLS recovery (reading B7) with ONE window that spans
// the whole loop and the dependency check answered by the profile (path 8).
//
// Reading B7 (P:L320-333 SE / DC / commit / mis-speculation
// recovery) runs fixed windows: every iteration speculates against the memory
// of the window start, DC marks the iterations with an exposed read written by
// an earlier iteration of the window, the violators are re-executed in
// dependence order with the operand forwarded from the writer's shadow slot,
// and the window commits whole.  Its statistics (jpo_sim_tls_fwd) only depend
// on W.  With W = n the windows -- and the grid barrier between them, ~45% of
// each window of the all-SM kernel -- disappear:
//
//   DC:       the violators of the one window are exactly the raw iterations
//             (an exposed read written by an earlier iteration of the loop);
//             the profile's guide (reading B5) already holds that bit, so no
//             write log is kept and nothing is probed;
//   SE:       a non-violator's exposed read is of an element no earlier
//             iteration writes; with write-once (waw = 0) and WAR-free
//             (war = 0) loops no LATER iteration writes it either, so its value
//             in A is the window-start value whenever it is read, and the
//             iteration's result is final: it commits in place at once;
//   recovery: a violator waits for its writer's shadow slot V[a] = 1 << 32 |
//             value (published by every RAW source, the guide's second
//             bitmap), then computes, commits, and publishes in turn.
//
// Iterations are dealt in slot sets (i = base + k*G + g) and taken in
// increasing order by every thread of a co-resident (cooperative) grid: the
// smallest unfinished iteration only waits for earlier, finished ones, so the
// sweep cannot deadlock.  Statistics are those of jpo_sim_tls_fwd with W = n:
// one window, violations = raw iterations, executed = n + violations.
// ADD_C only (one exposed read of A; configs 1, 3 and the config-5 middle).
#include <cooperative_groups.h>
#include "jp_host.h"

namespace cg = cooperative_groups;

namespace jp {

// CTA shape (measured on config 3, whole jp_schedule, d = 0.1/1/5/10%: 512 x 8 x 1
// CTA/SM 0.738/0.746/0.812/0.880 ms; 512 x 4 x 2 0.743/0.736/0.788/0.856; 1024 x 4
// 0.746/0.742/0.797/0.857; 256 x 8 x 3 0.770/0.778/0.865/0.947): random-access bound
#ifndef JP_FLOW_T
#define JP_FLOW_T 512
#endif
#ifndef JP_FLOW_K
#define JP_FLOW_K 4
#endif
#ifndef JP_FLOW_MINB
#define JP_FLOW_MINB 2
#endif
constexpr int kFlowT = JP_FLOW_T, kFlowK = JP_FLOW_K;
constexpr unsigned long long kFlowTag = 1ull << 32;
constexpr long long kFlowSpinLimit = 1ll << 22;   // a lost writer (inconsistent guide) ends the wait with an error

struct FlowSet {
  int32_t r[kFlowK], w[kFlowK];
  uint32_t gr[kFlowK], gs[kFlowK];
  uint32_t x[kFlowK];
};

template <int DT>
struct Flow {
  DLoop L;
  const uint32_t *graw, *gsrc;
  const uint32_t *o;     // ph: every non-violator's value, from k_flow_gath
  bool ph = false;
  unsigned long long *V;
  const int32_t *wsrc;   // nullable: writer of each raw iteration's read (loop-local id)
  uint32_t G, g, n, io, lo;
  uint32_t viol = 0;
  bool lost = false;

  __device__ __forceinline__ bool act(uint32_t base, int k) const { return base + (uint32_t)k * G + g < n; }
  __device__ __forceinline__ uint32_t it(uint32_t base, int k) const { return base + (uint32_t)k * G + g; }
  __device__ __forceinline__ bool raw_bit(const FlowSet &s, uint32_t base, int k) const {
    return (s.gr[k] >> (it(base, k) & 31)) & 1u;
  }
  __device__ __forceinline__ bool src_bit(const FlowSet &s, uint32_t base, int k) const {
    return (s.gs[k] >> (it(base, k) & 31)) & 1u;
  }
  __device__ __forceinline__ void load(uint32_t base, FlowSet &s) const {
#pragma unroll
    for (int k = 0; k < kFlowK; k++) {
      if (!act(base, k)) continue;
      const uint32_t i = it(base, k);
      s.w[k] = L.w ? __ldcs(L.w + i) : (int32_t)(io + i);
      s.gr[k] = __ldcs(graw + (i >> 5));
      s.gs[k] = __ldcs(gsrc + (i >> 5));
      if (ph) {   // the violators' read addresses; the others' values, gathered already
        if (raw_bit(s, base, k)) s.r[k] = L.r ? __ldcs(L.r + i) : (int32_t)(io + i);
        else s.x[k] = __ldcs(o + i);
      } else {
        s.r[k] = L.r ? __ldcs(L.r + i) : (int32_t)(io + i);
      }
    }
    if (wsrc) {   // a range of a loop: a raw read written before the range reads A
#pragma unroll
      for (int k = 0; k < kFlowK; k++)
        if (act(base, k) && raw_bit(s, base, k) && (uint32_t)__ldcs(wsrc + it(base, k)) < lo)
          s.gr[k] &= ~(1u << (it(base, k) & 31));
    }
  }
  // exposed reads of the non-violators (the violators' operands come from V)
  __device__ __forceinline__ void gather(uint32_t base, FlowSet &s) const {
    if (ph) return;
#pragma unroll
    for (int k = 0; k < kFlowK; k++)
      if (act(base, k) && !raw_bit(s, base, k)) s.x[k] = __ldcg(L.A + s.r[k]);
  }
  __device__ __forceinline__ void commit(const FlowSet &s, uint32_t base, int k, uint32_t v) const {
    __stcg(L.A + s.w[k], v);
    if (src_bit(s, base, k))
      asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(V + s.w[k]), "l"(kFlowTag | v) : "memory");
  }
  __device__ __forceinline__ void run(uint32_t base, FlowSet &s) {
    uint32_t pend = 0;
#pragma unroll
    for (int k = 0; k < kFlowK; k++) {
      if (!act(base, k)) continue;
      if (raw_bit(s, base, k)) pend |= 1u << k;
      else commit(s, base, k, ph ? s.x[k] : op_add<DT>(s.x[k], L.c0));
    }
    viol += __popc(pend);
    long long spins = 0;
    while (__any_sync(0xffffffffu, pend)) {
#pragma unroll
      for (int k = 0; k < kFlowK; k++) {
        if ((pend >> k) & 1u) {
          unsigned long long v;
          asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(V + s.r[k]) : "memory");
          if ((v >> 32) == 1ull) {
            commit(s, base, k, op_add<DT>((uint32_t)v, L.c0));
            pend &= ~(1u << k);
          }
        }
      }
      if (++spins > kFlowSpinLimit) {   // never on a consistent guide
        lost = lost || pend;
        break;
      }
    }
  }
};

template <int DT>
__global__ void __launch_bounds__(kFlowT, JP_FLOW_MINB) k_tls_flow(DLoop L, const uint32_t *graw, const uint32_t *gsrc,
                                                       unsigned long long *V, int64_t *stats, const int32_t *wsrc,
                                                       uint32_t lo, const int64_t *gate, int64_t raw_max,
                                                       const uint32_t *o, int64_t ph_max) {
  // gate (nullable): the profile header of this call -- launched before the host
  // has read it, the kernel runs only if the profile makes the loop a path-8 loop
  // (no bad index, war = waw = 0, 0 < raw <= raw_max, i.e. Fig. 2(b) mode B)
  if (gate && (gate[H_BAD] != 0 || gate[H_WAR] != 0 || gate[H_WAW] != 0 || gate[H_RAW] <= 0 || gate[H_RAW] > raw_max ||
               gate[H_GATE] != 0))
    return;
  Flow<DT> F;
  F.L = L; F.graw = graw; F.gsrc = gsrc; F.V = V; F.wsrc = wsrc; F.lo = lo;
  F.o = o;
  // the gather kernel ran ahead (k_flow_gath) exactly when the gate's raw count is at most ph_max
  F.ph = o && gate && gate[H_RAW] <= ph_max;
  F.G = gridDim.x * (uint32_t)kFlowT;
  F.g = blockIdx.x * (uint32_t)kFlowT + threadIdx.x;
  F.n = (uint32_t)L.n;
  F.io = (uint32_t)L.ioff;
  const uint32_t step = F.G * (uint32_t)kFlowK;
  // two slot sets in flight: the next set's indices, guide words and gathers
  // are issued before this set runs (a non-violator's operand is never written
  // by another iteration, so it may be read early)
  FlowSet a, b;
  F.load(0, a);
  F.gather(0, a);
  for (uint32_t base = 0; base < F.n; base += 2 * step) {
    if (base + step < F.n) { F.load(base + step, b); F.gather(base + step, b); }
    F.run(base, a);
    if (base + step >= F.n) break;
    if (base + 2 * step < F.n) { F.load(base + 2 * step, a); F.gather(base + 2 * step, a); }
    F.run(base + step, b);
  }
  const uint32_t v = __reduce_add_sync(0xffffffffu, F.viol);
  const unsigned lost = __any_sync(0xffffffffu, F.lost);
  if ((threadIdx.x & 31) == 0) {
    if (v) atomicAdd(reinterpret_cast<unsigned long long *>(&stats[3]), (unsigned long long)v);
    if (lost) atomicAdd(reinterpret_cast<unsigned long long *>(&stats[1]), 1ull);
  }
}

// The gather kernel of the phased sweep: o[i] = A[r[i]] + c0 for every
// non-violator (its operand is never written, B12), gated like the sweep on the
// profile header, plus raw <= ph_max.  2048 threads per SM (the sweep's register
// budget allows 1024): the gathers at the device's random-read rate.
template <int DT>
__global__ void __launch_bounds__(256) k_flow_gath(DLoop L, const uint32_t *graw, uint32_t *o, const int64_t *gate,
                                                   int64_t raw_max, int64_t ph_max) {
  if (gate[H_BAD] != 0 || gate[H_WAR] != 0 || gate[H_WAW] != 0 || gate[H_RAW] <= 0 || gate[H_RAW] > raw_max ||
      gate[H_GATE] != 0 || gate[H_RAW] > ph_max)
    return;
  constexpr int Q = 4;
  const int64_t G = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i0 = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i0 < L.n; i0 += G * Q) {
    int32_t r[Q];
    uint32_t raw[Q], x[Q];
#pragma unroll
    for (int u = 0; u < Q; u++) {
      const int64_t i = i0 + u * G;
      raw[u] = 1;
      if (i >= L.n) continue;
      raw[u] = (__ldcs(graw + (i >> 5)) >> (i & 31)) & 1u;
      r[u] = L.r ? __ldcs(L.r + i) : (int32_t)(L.ioff + i);
    }
#pragma unroll
    for (int u = 0; u < Q; u++)
      if (!raw[u]) x[u] = __ldcg(L.A + r[u]);
#pragma unroll
    for (int u = 0; u < Q; u++)
      if (!raw[u]) __stcs(o + i0 + u * G, op_add<DT>(x[u], L.c0));
  }
}

template <int DT>
static cudaError_t run_flow_gath(const Job &j, const uint32_t *graw, uint32_t *o, const int64_t *gate, int64_t raw_max,
                                 int64_t ph_max, cudaStream_t st) {
  int64_t cap = (int64_t)num_sms() * 8;
  const int64_t need = (j.d.n + 255) / 256;
  const int grid = (int)(need < 1 ? 1 : need < cap ? need : cap);
  k_flow_gath<DT><<<grid, 256, 0, st>>>(j.d, graw, o, gate, raw_max, ph_max);
  note_launch();
  return cudaSuccess;
}

template <int DT>
static cudaError_t run_flow(const Job &j, const uint32_t *graw, const uint32_t *gsrc, unsigned long long *V,
                            int64_t *stats, cudaStream_t st, const int32_t *wsrc, uint32_t lo, const int64_t *gate,
                            int64_t raw_max, int max_ctas, const uint32_t *o, int64_t ph_max) {
  static int maxb = 0;   // (one device model per process: B200)
  if (maxb < 1) cudaOccupancyMaxActiveBlocksPerMultiprocessor(&maxb, (const void *)k_tls_flow<DT>, kFlowT, 0);
  if (maxb < 1) return cudaErrorInvalidConfiguration;
  int grid = num_sms() * maxb;
  if (max_ctas > 0 && grid > max_ctas) grid = max_ctas;
  const int64_t need = (j.d.n + kFlowT - 1) / kFlowT;
  if (need < grid) grid = (int)(need < 1 ? 1 : need);
  DLoop d = j.d;
  void *args[] = {&d, &graw, &gsrc, &V, &stats, &wsrc, &lo, &gate, &raw_max, &o, &ph_max};
  note_launch();
  return cudaLaunchCooperativeKernel((const void *)k_tls_flow<DT>, dim3(grid), dim3(kFlowT), args, 0, st);
}

// ---------------------------------------------------------------------------
// Path 9 (reading B14): the same one window over a loop WITH WAR / WAW.  What
// changes against path 8:
//   recovery: the writer a violator must see is the LAST earlier writer of its
//             address, pred(i) (the profile's last-writer pass records it), and
//             its shadow slot is per ITERATION (V[pred]), since an address has
//             several values over the loop;
//   SE:       a non-violator's exposed read is of an element no earlier
//             iteration writes -- but a later one may (WAR): nothing writes A
//             in place except an address's last writer, and the last writer of
//             an address that has such an exposed read waits for the window's
//             one grid barrier (`later`); every other last writer (`now`)
//             commits at once -- no exposed read of its address exists, and
//             every other read of it is a violator fed from V;
//   commit:   the final value of an address is its last writer's (WAW order),
//             exactly the sequential state; writers that are not last only
//             publish (if some violator reads them).
// Statistics: jpo_sim_tls_fwd with W = n, as path 8.
// ---------------------------------------------------------------------------
struct FlowSetW {
  int32_t r[kFlowK], w[kFlowK], pr[kFlowK];
  uint32_t f[kFlowK];   // the iteration's bits: raw 1, publish 2, commit now 4, commit later 8
  uint32_t x[kFlowK];   // the exposed read of A (non-violators): A[r] (ADD_C), Y[w] (SAXPY)
  uint32_t xs[kFlowK];  // SAXPY: X[r] (read-only, gathered for every iteration)
};
constexpr uint32_t kFRaw = 1, kFPub = 2, kFNow = 4, kFLater = 8;

// OP: ADD_C (A[w] = A[r] + c0) or SAXPY (Y[w] = c0*X[r] + Y[w], its exposed read
// is of the address it writes: a scatter-add whose duplicate writes chain)
template <int OP, int DT>
struct FlowW {
  DLoop L;
  const uint32_t *graw, *gpub, *gnow, *glater;
  const int32_t *pred;
  unsigned long long *V;
  uint32_t G, g, n, io;
  uint32_t viol = 0;
  bool lost = false;

  __device__ __forceinline__ bool act(uint32_t base, int k) const { return base + (uint32_t)k * G + g < n; }
  __device__ __forceinline__ uint32_t it(uint32_t base, int k) const { return base + (uint32_t)k * G + g; }
  __device__ __forceinline__ void load(uint32_t base, FlowSetW &s) const {
#pragma unroll
    for (int k = 0; k < kFlowK; k++) {
      s.f[k] = 0;
      if (!act(base, k)) continue;
      const uint32_t i = it(base, k), q = i >> 5, sh = i & 31;
      s.r[k] = L.r ? __ldcs(L.r + i) : (int32_t)(io + i);
      s.w[k] = L.w ? __ldcs(L.w + i) : (int32_t)(io + i);
      s.f[k] = ((__ldcs(graw + q) >> sh) & 1u) | ((__ldcs(gpub + q) >> sh) & 1u) << 1 |
               ((__ldcs(gnow + q) >> sh) & 1u) << 2 | ((__ldcs(glater + q) >> sh) & 1u) << 3;
    }
#pragma unroll
    for (int k = 0; k < kFlowK; k++)
      if (s.f[k] & kFRaw) s.pr[k] = __ldcs(pred + it(base, k));
  }
  __device__ __forceinline__ void gather(uint32_t base, FlowSetW &s) const {
#pragma unroll
    for (int k = 0; k < kFlowK; k++) {
      if (!act(base, k)) continue;
      if constexpr (OP == JP_OP_SAXPY) s.xs[k] = __ldcg(L.X + s.r[k]);
      if (!(s.f[k] & kFRaw)) s.x[k] = __ldcg(L.A + (OP == JP_OP_SAXPY ? s.w[k] : s.r[k]));
    }
  }
  // the body's value from the exposed read a (of A / Y)
  __device__ __forceinline__ uint32_t body(const FlowSetW &s, int k, uint32_t a) const {
    if constexpr (OP == JP_OP_SAXPY) return op_add<DT>(op_mul<DT>(L.c0, s.xs[k]), a);
    else return op_add<DT>(a, L.c0);
  }
  __device__ __forceinline__ void commit(const FlowSetW &s, uint32_t base, int k, uint32_t v) const {
    if (s.f[k] & kFNow) __stcg(L.A + s.w[k], v);
    if (s.f[k] & (kFPub | kFLater))
      asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(V + it(base, k)), "l"(kFlowTag | v) : "memory");
  }
  __device__ __forceinline__ void run(uint32_t base, FlowSetW &s) {
    uint32_t pend = 0;
#pragma unroll
    for (int k = 0; k < kFlowK; k++) {
      if (!act(base, k)) continue;
      if (s.f[k] & kFRaw) pend |= 1u << k;
      else commit(s, base, k, body(s, k, s.x[k]));
    }
    viol += __popc(pend);
    long long spins = 0;
    while (__any_sync(0xffffffffu, pend)) {
#pragma unroll
      for (int k = 0; k < kFlowK; k++) {
        if ((pend >> k) & 1u) {
          unsigned long long v;
          asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(V + s.pr[k]) : "memory");
          if ((v >> 32) == 1ull) {
            commit(s, base, k, body(s, k, (uint32_t)v));
            pend &= ~(1u << k);
          }
        }
      }
      if (++spins > kFlowSpinLimit) {
        lost = lost || pend;
        break;
      }
    }
  }
};

template <int OP, int DT>
__global__ void __launch_bounds__(kFlowT, JP_FLOW_MINB) k_tls_flow_waw(DLoop L, const uint32_t *graw, const int32_t *pred,
                                                           const uint32_t *bits, unsigned long long *V,
                                                           int64_t *stats, const int64_t *gate) {
  if (gate && gate[H_PRED_FAIL] != 0) return;   // grid-uniform: no barrier is entered
  const uint32_t nw = (uint32_t)((L.n + 31) / 32);
  FlowW<OP, DT> F;
  F.L = L; F.graw = graw; F.pred = pred; F.V = V;
  F.gpub = bits; F.gnow = bits + nw; F.glater = bits + 2 * nw;
  F.G = gridDim.x * (uint32_t)kFlowT;
  F.g = blockIdx.x * (uint32_t)kFlowT + threadIdx.x;
  F.n = (uint32_t)L.n;
  F.io = (uint32_t)L.ioff;
  const uint32_t step = F.G * (uint32_t)kFlowK;
  FlowSetW a, b;
  F.load(0, a);
  F.gather(0, a);
  for (uint32_t base = 0; base < F.n; base += 2 * step) {
    if (base + step < F.n) { F.load(base + step, b); F.gather(base + step, b); }
    F.run(base, a);
    if (base + step >= F.n) break;
    if (base + 2 * step < F.n) { F.load(base + 2 * step, a); F.gather(base + 2 * step, a); }
    F.run(base + step, b);
  }
  const uint32_t v = __reduce_add_sync(0xffffffffu, F.viol);
  const unsigned lost = __any_sync(0xffffffffu, F.lost);
  if ((threadIdx.x & 31) == 0) {
    if (v) atomicAdd(reinterpret_cast<unsigned long long *>(&stats[3]), (unsigned long long)v);
    if (lost) atomicAdd(reinterpret_cast<unsigned long long *>(&stats[1]), 1ull);
  }
  // the window's one barrier: then the last writers whose address had an exposed
  // read (its window-start value is no longer needed) commit from their slots
  cg::this_grid().sync();
  for (uint32_t q = F.g; q < nw; q += F.G) {
    uint32_t m = __ldcs(F.glater + q);
    while (m) {
      const uint32_t i = q * 32 + (uint32_t)__ffs(m) - 1;
      m &= m - 1;
      const int32_t wi = L.w ? L.w[i] : (int32_t)(F.io + i);
      L.A[wi] = (uint32_t)__ldcg(V + i);
    }
  }
}

template <int OP, int DT>
static cudaError_t run_flow_waw(const Job &j, const uint32_t *graw, const int32_t *pred, const uint32_t *bits,
                                unsigned long long *V, int64_t *stats, const int64_t *gate, cudaStream_t st) {
  static int maxb = 0;   // (one device model per process: B200)
  if (maxb < 1) cudaOccupancyMaxActiveBlocksPerMultiprocessor(&maxb, (const void *)k_tls_flow_waw<OP, DT>, kFlowT, 0);
  if (maxb < 1) return cudaErrorInvalidConfiguration;
  int grid = num_sms() * maxb;
  const int64_t need = (j.d.n + kFlowT - 1) / kFlowT;
  if (need < grid) grid = (int)(need < 1 ? 1 : need);
  DLoop d = j.d;
  void *args[] = {&d, &graw, &pred, &bits, &V, &stats, &gate};
  note_launch();
  return cudaLaunchCooperativeKernel((const void *)k_tls_flow_waw<OP, DT>, dim3(grid), dim3(kFlowT), args, 0, st);
}

cudaError_t launch_tls_flow_waw(const Job &j, const uint32_t *graw, const int32_t *pred, const uint32_t *bits,
                                unsigned long long *V, int64_t *stats, const int64_t *gate, cudaStream_t st) {
  cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
  if (j.d.n == 0) return launch_check();
  cudaError_t e;
  if (j.op == JP_OP_ADD_C)
    e = j.dt == JP_F32 ? run_flow_waw<JP_OP_ADD_C, JP_F32>(j, graw, pred, bits, V, stats, gate, st)
                       : run_flow_waw<JP_OP_ADD_C, JP_I32>(j, graw, pred, bits, V, stats, gate, st);
  else if (j.op == JP_OP_SAXPY)
    e = j.dt == JP_F32 ? run_flow_waw<JP_OP_SAXPY, JP_F32>(j, graw, pred, bits, V, stats, gate, st)
                       : run_flow_waw<JP_OP_SAXPY, JP_I32>(j, graw, pred, bits, V, stats, gate, st);
  else
    return cudaErrorInvalidValue;
  if (e != cudaSuccess) return e;
  return launch_check();
}

// Device stats after the kernel: stats[3] = violations (raw iterations),
// stats[1] = number of warps that gave up waiting for a writer (0 unless the
// guide was inconsistent); the caller turns them into jpo_sim_tls_fwd's
// (committed n, executed n + violations, windows 1).  V must hold no value
// tagged 1 << 32 for an address the loop writes (zeroed).
cudaError_t launch_tls_flow(const Job &j, const uint32_t *graw, const uint32_t *gsrc, unsigned long long *V,
                            int64_t *stats, cudaStream_t st, const int32_t *wsrc, int64_t lo, const int64_t *gate,
                            int64_t raw_max, bool zero_stats, int max_ctas, uint32_t *o, int64_t ph_max) {
  if (zero_stats) cudaMemsetAsync(stats, 0, 4 * sizeof(int64_t), st);
  if (j.d.n == 0) return launch_check();
  if (j.op != JP_OP_ADD_C) return cudaErrorInvalidValue;
  // o with a gate: the non-violators' values gathered by a kernel of their own
  // first (all the loop's random reads ahead of its writes: B200's L2 serves them
  // faster apart, scripts/ubench/rand_phase.cu), when the gate's raw count is at
  // most ph_max (few violators: the sweep then hardly waits)
  const char *pe = getenv("JP_FLOW_PHASED");
  if (!gate || (pe && pe[0] == '0')) o = nullptr;
  cudaError_t e = cudaSuccess;
  if (o) e = j.dt == JP_F32 ? run_flow_gath<JP_F32>(j, graw, o, gate, raw_max, ph_max, st)
                            : run_flow_gath<JP_I32>(j, graw, o, gate, raw_max, ph_max, st);
  if (e != cudaSuccess) return e;
  e = j.dt == JP_F32 ? run_flow<JP_F32>(j, graw, gsrc, V, stats, st, wsrc, (uint32_t)lo, gate, raw_max, max_ctas, o, ph_max)
                     : run_flow<JP_I32>(j, graw, gsrc, V, stats, st, wsrc, (uint32_t)lo, gate, raw_max, max_ctas, o, ph_max);
  if (e != cudaSuccess) return e;
  return launch_check();
}

}  // namespace jp

// jp_profile.cu -- dependency-density profiler kernels (Fig. 1 "Profiler / DD
// analysis, intra-warp / inter-warp").
//
// Pass 1 (stamp): every access a of iteration gid stamps the per-array tables
//   minW[a] (writes) and minR[a] (exposed + covered reads) with the earliest gid,
//   encoded INT32_MAX - gid so that atomicMax == earliest and an int32 MAX
//   all-reduce composes ranks (C1).  Out-of-range indices are counted (fused
//   validation, reading A13) and skipped.  Small arrays (<= 4096 elements, the
//   private(list) scratch of config 4) are pre-aggregated in shared memory
//   with a check-before-atomic filter; ascending gid order inside a CTA makes
//   every touch after the first a no-op.
// Pass 2 (classify): per iteration raw/war/waw against the tables (reading
//   A1).  Counts only (jp_schedule's call): per-thread counters, one warp
//   reduction and one global atomic per CTA.  With a raw bitmap (D4) or
//   per-chunk counts: __ballot_sync + __popc per warp tile of 32 iterations.
// Both passes take 4 consecutive iterations per thread (16-byte index loads)
// with two steps in flight and 32-bit index arithmetic.
// The intra-warp / inter-warp split of the paper is an
// implementation detail here (reading A2): results do not depend on geometry.
#include <cstdlib>
#include "jp_host.h"

namespace jp {

// table bytes stamped per pass (env JP_STAMP_PASS_MB overrides, for measurement)
// env knob read per call (tests and measurements flip it), default dflt
static int getenv_int(const char *name, int dflt) {
  const char *e = getenv(name);
  return e && e[0] ? atoi(e) : dflt;
}

static size_t stamp_pass_bytes() {
  const char *e = getenv("JP_STAMP_PASS_MB");
  const long mb = e ? atol(e) : 48;
  return (size_t)(mb > 0 ? mb : 48) << 20;
}

struct Tabs {
  int32_t *wA, *rA, *wT, *rT;
  // optional interleaved copy {minW[a], minR[a]} of the A tables (classify only):
  // the war and waw lookups of a written address then cost one 8-byte access
  // (one DRAM burst) instead of two in separate 64 MiB tables
  const int2 *pA;
  int as;   // element stride of wA / rA (1; 2 when they point into the pairs)
  int sA, sT;   // pre-aggregate in shared memory
  // stamp pass over an address window [lo, lo + span) only (tables larger than
  // L2 are stamped in several passes, each with an L2-resident working set);
  // index errors are counted by the pass with count_bad
  uint32_t lo, span;
  int count_bad;
};

__device__ __forceinline__ void check(int64_t a, int64_t len, int64_t &bad) {
  if ((uint64_t)a >= (uint64_t)len) bad++;
}

// Loads of kUnroll iterations (one per CTA-wide slice) are issued before any
// of them is used: the passes stream their index arrays from HBM, and one
// dependent load chain per warp at a time would leave them latency-bound.
constexpr int kUnroll = 4;

// ---------------------------------------------------------------------------
// Quad variants: each thread takes 4 consecutive iterations per step (one
// 16-byte load per index stream when every stream is 16-byte aligned), two
// steps in flight, 32-bit index arithmetic.  Same tables, same counts.
// ---------------------------------------------------------------------------
__device__ __forceinline__ int4 idx4(const DLoop &L, const int32_t *p, int64_t i, bool vec) {
  if (!p) {
    const int b = (int)(L.ioff + i);
    return make_int4(b, b + 1, b + 2, b + 3);
  }
  if (vec && i + 4 <= L.n) return __ldcs(reinterpret_cast<const int4 *>(p + i));
  int4 r;
  r.x = p[i];
  r.y = i + 1 < L.n ? p[i + 1] : 0;
  r.z = i + 2 < L.n ? p[i + 2] : 0;
  r.w = i + 3 < L.n ? p[i + 3] : 0;
  return r;
}
__device__ __forceinline__ int q4(const int4 &v, int k) { return k == 0 ? v.x : k == 1 ? v.y : k == 2 ? v.z : v.w; }
// chk: the index came from an index array (identity indices were range-checked on the host)
// gs: element stride of the global table (2 when the A tables are stamped
// straight into interleaved {minW, minR} pairs, jp_schedule)
__device__ __forceinline__ void stamp32(int32_t *g, int32_t *s, int32_t a, int32_t len, int32_t e, const Tabs &t,
                                        int &bad, bool chk = true, int gs = 1) {
  if (chk && (uint32_t)a >= (uint32_t)len) { bad += t.count_bad; return; }
  if ((uint32_t)a - t.lo >= t.span) return;
  if (s) {
    if (s[a] < e) atomicMax(&s[a], e);
  } else if (g) {
    atomicMax(&g[(int64_t)a * gs], e);
  }
}
__device__ __forceinline__ bool earlier32(const int32_t *tab, int32_t a, int32_t len, int32_t e) {
  return tab && (uint32_t)a < (uint32_t)len && tab[a] > e;
}
constexpr int kQuadSteps = 2;

template <int OP>
__global__ void __launch_bounds__(256) k_prof_stamp4(DLoop L, Tabs t, int vec, int64_t *hdr) {
  extern __shared__ int32_t sm[];
  int32_t *sAw = nullptr, *sAr = nullptr, *sTw = nullptr;
  int32_t *p = sm;
  if (t.sA) { sAw = p; p += L.lenA; if (t.rA) { sAr = p; p += L.lenA; } }
  if (t.sT) { sTw = p; p += L.lenT; }   // minR(T) == minW(T) for PRIV_TMP (see k_prof_stamp)
  for (int64_t k = threadIdx.x; k < p - sm; k += blockDim.x) sm[k] = -1;
  JP_CTA_SYNC();
  const int32_t lenA = (int32_t)L.lenA, lenX = (int32_t)L.lenX, lenT = (int32_t)L.lenT;
  const bool hr = L.r != nullptr, hw = L.w != nullptr,
             h2 = (OP == JP_OP_STENCIL2 ? L.r2 : OP == JP_OP_PRIV_TMP ? L.s : nullptr) != nullptr;
  int bad = 0;
  const int64_t nq = (L.n + 3) >> 2, B = blockDim.x;
  for (int64_t q0 = (int64_t)blockIdx.x * B * kQuadSteps + threadIdx.x; q0 < nq; q0 += (int64_t)gridDim.x * B * kQuadSteps) {
    int4 va[kQuadSteps], vb[kQuadSteps], vc[kQuadSteps];
#pragma unroll
    for (int u = 0; u < kQuadSteps; u++) {
      const int64_t q = q0 + u * B;
      if (q < nq) {
        const int64_t i = q << 2;
        if constexpr (OP == JP_OP_ADD_C || OP == JP_OP_SAXPY) { va[u] = idx4(L, L.w, i, vec); vb[u] = idx4(L, L.r, i, vec); }
        else if constexpr (OP == JP_OP_PRIV_TMP) { va[u] = idx4(L, L.s, i, vec); vb[u] = idx4(L, L.r, i, vec); vc[u] = idx4(L, L.w, i, vec); }
        else { va[u] = idx4(L, L.w, i, vec); vb[u] = idx4(L, L.r, i, vec); vc[u] = idx4(L, L.r2, i, vec); }
      }
    }
#pragma unroll
    for (int u = 0; u < kQuadSteps; u++) {
      const int64_t q = q0 + u * B;
      if (q >= nq) break;
      const int32_t e0 = enc_gid(L.base + (q << 2));
      const int kn = L.n - (q << 2) < 4 ? (int)(L.n - (q << 2)) : 4;
#pragma unroll
      for (int k = 0; k < 4; k++) {
        if (k >= kn) break;
        const int32_t e = e0 - k;
        const int32_t a = q4(va[u], k), b = q4(vb[u], k);
        // identity streams (NULL arrays) were range-checked on the host and
        // reach a table only when the array is also reached through an index
        if constexpr (OP == JP_OP_ADD_C) {
          stamp32(t.wA, sAw, a, lenA, e, t, bad, hw, t.as);
          stamp32(t.rA, sAr, b, lenA, e, t, bad, hr, t.as);
        } else if constexpr (OP == JP_OP_SAXPY) {
          if (hr && (uint32_t)b >= (uint32_t)lenX) bad++;
          if (hw) {
            stamp32(t.wA, sAw, a, lenA, e, t, bad, true, t.as);
            if ((uint32_t)a < (uint32_t)lenA) stamp32(t.rA, sAr, a, lenA, e, t, bad, false, t.as);
          }
        } else if constexpr (OP == JP_OP_PRIV_TMP) {
          if (hr && (uint32_t)b >= (uint32_t)lenX) bad++;
          if (h2) {
            if (sTw) {
              stamp32(t.wT, sTw, a, lenT, e, t, bad);
            } else {
              stamp32(t.wT, nullptr, a, lenT, e, t, bad);
              if ((uint32_t)a < (uint32_t)lenT) stamp32(t.rT, nullptr, a, lenT, e, t, bad, false);
            }
          }
          if (hw) stamp32(t.wA, sAw, q4(vc[u], k), lenA, e, t, bad, true, t.as);
        } else {
          stamp32(t.wA, sAw, a, lenA, e, t, bad, hw, t.as);
          stamp32(t.rA, sAr, b, lenA, e, t, bad, hr, t.as);
          stamp32(t.rA, sAr, q4(vc[u], k), lenA, e, t, bad, h2, t.as);
        }
      }
    }
  }
  bad = __reduce_add_sync(0xffffffffu, bad);
  if ((threadIdx.x & 31) == 0 && bad) atomicAdd((unsigned long long *)&hdr[H_BAD], (unsigned long long)bad);
  JP_CTA_SYNC();
  if (t.sA) {
    for (int64_t a = threadIdx.x; a < L.lenA; a += blockDim.x) {
      if (sAw[a] != -1) atomicMax(&t.wA[a], sAw[a]);
      if (sAr && sAr[a] != -1) atomicMax(&t.rA[a], sAr[a]);
    }
  }
  if (t.sT) {
    for (int64_t a = threadIdx.x; a < L.lenT; a += blockDim.x)
      if (sTw[a] != -1) { atomicMax(&t.wT[a], sTw[a]); atomicMax(&t.rT[a], sTw[a]); }
  }
}

// counts-only classify (no raw bitmap, no chunk counts): per-thread counters,
// one reduction per CTA.  GUIDE: also the TLS guide bitmaps of jp_tls_guide
// (region 13) in the same pass -- raw words by an OR over the 8 lanes that
// share a word, and RAW-source words by an atomicOr at each raw read's first
// writer.  The source words equal jp_tls_guide's whenever the loop writes no
// address twice (then an address read by a later iteration has exactly one
// writer, the first), which is the only case a guided TLS run accepts; the
// caller zeroes them first.
__device__ __forceinline__ int2 pair32(const int2 *p, int32_t a, int32_t len) {
  return (uint32_t)a < (uint32_t)len ? __ldg(p + a) : make_int2(-1, -1);
}

// cc (nullable): per-chunk raw / war / waw counts, chunk % 32 == 0 and >= 128,
// so a warp's 128 consecutive iterations of one quad step span at most two chunks
template <int OP, bool GUIDE, bool PAIRS = false>
__global__ void __launch_bounds__(256) k_prof_count4(DLoop L, Tabs t, int vec, int64_t *hdr, uint32_t *graw,
                                                     uint32_t *gsrc, int64_t chunk = 0, int64_t *cc = nullptr,
                                                     unsigned long long *dist = nullptr) {
  __shared__ unsigned long long s_cnt[3];
  __shared__ unsigned long long s_first;
  // PRIV_TMP with a small T (config 4: 1024 slots): its first-writer table in
  // shared memory -- a warp's 32 random slot lookups would otherwise be up to
  // 32 L1 wavefronts per load
  __shared__ int32_t s_tT[OP == JP_OP_PRIV_TMP ? kSmemSlots : 1];
  if (threadIdx.x < 3) s_cnt[threadIdx.x] = 0;
  if (threadIdx.x == 0) s_first = ~0ull;
  const int32_t lenA = (int32_t)L.lenA, lenT = (int32_t)L.lenT;
  const int32_t *wT = t.wT;
  if constexpr (OP == JP_OP_PRIV_TMP) {
    if (t.wT && lenT <= kSmemSlots) {
      for (int k = threadIdx.x; k < lenT; k += blockDim.x) s_tT[k] = __ldg(t.wT + k);
      wT = s_tT;
    }
  }
  JP_CTA_SYNC();
  const int32_t *rT = OP == JP_OP_PRIV_TMP ? wT : t.rT;
  unsigned c_raw = 0, c_war = 0, c_waw = 0;
  unsigned long long first = ~0ull;
  const int64_t nq = (L.n + 3) >> 2, B = blockDim.x;
  // the writer (local iteration) behind a raw read of address a: mark it a RAW
  // source, and count the read's dependence distance i - j (floor log2) for the
  // restart-TLS window choice (jp_schedule, restart_plan)
  __shared__ unsigned s_dist[GUIDE ? 32 : 1];
  if (GUIDE && threadIdx.x < 32) s_dist[threadIdx.x] = 0;
  auto mark_src = [&](int32_t a, int32_t e) {
    if constexpr (GUIDE) {
      const int32_t we = PAIRS ? t.pA[a].x : t.wA[a];
      const int64_t j = (int64_t)(0x7FFFFFFF - we) - L.base;
      atomicOr(&gsrc[j >> 5], 1u << (j & 31));
      if (dist) atomicAdd(&s_dist[31 - __clz(we - e)], 1u);
    }
  };
  for (int64_t q0 = (int64_t)blockIdx.x * B * kQuadSteps + threadIdx.x; q0 - threadIdx.x < nq; q0 += (int64_t)gridDim.x * B * kQuadSteps) {
    int4 va[kQuadSteps], vb[kQuadSteps], vc[kQuadSteps];
#pragma unroll
    for (int u = 0; u < kQuadSteps; u++) {
      const int64_t q = q0 + u * B;
      if (q < nq) {
        const int64_t i = q << 2;
        if constexpr (OP == JP_OP_ADD_C) { va[u] = idx4(L, L.w, i, vec); vb[u] = idx4(L, L.r, i, vec); }
        else if constexpr (OP == JP_OP_SAXPY) { va[u] = idx4(L, L.w, i, vec); }
        else if constexpr (OP == JP_OP_PRIV_TMP) { va[u] = idx4(L, L.s, i, vec); vb[u] = idx4(L, L.w, i, vec); }
        else { va[u] = idx4(L, L.w, i, vec); vb[u] = idx4(L, L.r, i, vec); vc[u] = idx4(L, L.r2, i, vec); }
      }
    }
#pragma unroll
    for (int u = 0; u < kQuadSteps; u++) {
      const int64_t q = q0 + u * B;
      uint32_t rb = 0;   // raw bits of this lane's 4 iterations
      unsigned qr = 0, qa = 0, qw = 0;   // this quad's counts (chunk counts)
      if (q < nq) {
        const int32_t e0 = enc_gid(L.base + (q << 2));
        const int kn = L.n - (q << 2) < 4 ? (int)(L.n - (q << 2)) : 4;
#pragma unroll
        for (int k = 0; k < 4; k++) {
          if (k >= kn) break;
          const int32_t e = e0 - k;
          const int32_t a = q4(va[u], k);
          bool raw = false, war, waw;
          if constexpr (OP == JP_OP_ADD_C) {
            // r == w (an in-place update, most iterations of configs 3 and 5):
            // the raw and waw lookups are the same table entry -- one load
            const int32_t b = q4(vb[u], k);
            if constexpr (PAIRS) {
              const int2 pa = pair32(t.pA, a, lenA);
              war = pa.y > e;
              waw = pa.x > e;
            } else {
              war = earlier32(t.rA, a, lenA, e);
              waw = earlier32(t.wA, a, lenA, e);
            }
            raw = b == a ? waw : PAIRS ? pair32(t.pA, b, lenA).x > e : earlier32(t.wA, b, lenA, e);
            if (raw) mark_src(b, e);
          } else if constexpr (OP == JP_OP_SAXPY) {
            if constexpr (PAIRS) {
              const int2 pa = pair32(t.pA, a, lenA);
              raw = pa.x > e;
              war = pa.y > e;
            } else {
              raw = earlier32(t.wA, a, lenA, e);
              war = earlier32(t.rA, a, lenA, e);
            }
            waw = raw;
            if (raw) mark_src(a, e);
          } else if constexpr (OP == JP_OP_PRIV_TMP) {
            war = earlier32(rT, a, lenT, e);
            waw = earlier32(wT, a, lenT, e) || earlier32(t.wA, q4(vb[u], k), lenA, e);
          } else {
            if constexpr (PAIRS) {
              const int2 pa = pair32(t.pA, a, lenA);
              war = pa.y > e;
              waw = pa.x > e;
            } else {
              war = earlier32(t.rA, a, lenA, e);
              waw = earlier32(t.wA, a, lenA, e);
            }
            const int32_t b = q4(vb[u], k), c = q4(vc[u], k);
            const bool r0 = b == a ? waw : PAIRS ? pair32(t.pA, b, lenA).x > e : earlier32(t.wA, b, lenA, e);
            const bool r1 = c == a ? waw : c == b ? r0 : PAIRS ? pair32(t.pA, c, lenA).x > e : earlier32(t.wA, c, lenA, e);
            raw = r0 || r1;
            if (r0) mark_src(q4(vb[u], k), e);
            if (r1) mark_src(q4(vc[u], k), e);
          }
          c_raw += raw; c_war += war; c_waw += waw;
          qr += raw; qa += war; qw += waw;
          rb |= (uint32_t)raw << k;
          if (raw && first == ~0ull) first = (unsigned long long)(L.base + (q << 2) + k);
        }
      }
      if (cc && q0 - threadIdx.x + u * B < nq) {   // warp-uniform: some lane of the warp has a quad
        const int64_t c = q < nq ? (q << 2) / chunk : -1;
        const int64_t c0 = __shfl_sync(0xffffffffu, c, 0);
        const bool in0 = c == c0;
        const unsigned r0 = __reduce_add_sync(0xffffffffu, in0 ? qr : 0u), r1 = __reduce_add_sync(0xffffffffu, in0 ? 0u : qr);
        const unsigned a0 = __reduce_add_sync(0xffffffffu, in0 ? qa : 0u), a1 = __reduce_add_sync(0xffffffffu, in0 ? 0u : qa);
        const unsigned w0 = __reduce_add_sync(0xffffffffu, in0 ? qw : 0u), w1 = __reduce_add_sync(0xffffffffu, in0 ? 0u : qw);
        const int64_t c1 = __reduce_max_sync(0xffffffffu, (unsigned)(c < 0 ? 0 : c));
        if ((threadIdx.x & 31) == 0) {
          auto add = [&](int64_t ch, int kind, unsigned v) {
            if (v) atomicAdd(reinterpret_cast<unsigned long long *>(&cc[3 * ch + kind]), (unsigned long long)v);
          };
          add(c0, 0, r0); add(c0, 1, a0); add(c0, 2, w0);
          if (c1 != c0) { add(c1, 0, r1); add(c1, 1, a1); add(c1, 2, w1); }
        }
      }
      if constexpr (GUIDE) {
        // lanes 8m..8m+7 hold the 32 iterations of one word (q0 of lane 0 is a multiple of 8)
        uint32_t wv = rb << (4 * (threadIdx.x & 7));
        wv |= __shfl_xor_sync(0xffffffffu, wv, 1);
        wv |= __shfl_xor_sync(0xffffffffu, wv, 2);
        wv |= __shfl_xor_sync(0xffffffffu, wv, 4);
        if ((threadIdx.x & 7) == 0 && q < nq) graw[q >> 3] = wv;
      }
    }
  }
  c_raw = __reduce_add_sync(0xffffffffu, c_raw);
  c_war = __reduce_add_sync(0xffffffffu, c_war);
  c_waw = __reduce_add_sync(0xffffffffu, c_waw);
  for (int o = 16; o; o >>= 1) {
    const unsigned long long x = __shfl_xor_sync(0xffffffffu, first, o);
    first = x < first ? x : first;
  }
  if ((threadIdx.x & 31) == 0) {
    if (c_raw) atomicAdd(&s_cnt[0], (unsigned long long)c_raw);
    if (c_war) atomicAdd(&s_cnt[1], (unsigned long long)c_war);
    if (c_waw) atomicAdd(&s_cnt[2], (unsigned long long)c_waw);
    if (first != ~0ull) atomicMin(&s_first, first);
  }
  JP_CTA_SYNC();
  if (threadIdx.x < 3 && s_cnt[threadIdx.x]) atomicAdd((unsigned long long *)&hdr[H_RAW + threadIdx.x], s_cnt[threadIdx.x]);
  if (threadIdx.x == 0 && s_first != ~0ull) atomicMin((unsigned long long *)&hdr[H_FIRST_RAW], s_first);
  if constexpr (GUIDE) {
    if (dist && threadIdx.x < 32 && s_dist[threadIdx.x]) atomicAdd(&dist[threadIdx.x], (unsigned long long)s_dist[threadIdx.x]);
  }
}

static int idx_vec(const DLoop &d) {
  auto al = [](const int32_t *q) { return q == nullptr || ((uintptr_t)q & 15) == 0; };
  return al(d.r) && al(d.w) && al(d.r2) && al(d.s);
}

// (bounds-guarded: classify may run before the host has seen the bad-index count)
__device__ __forceinline__ bool earlier(const int32_t *tab, int64_t a, int64_t len, int32_t e, int stride = 1) {
  return tab && (uint64_t)a < (uint64_t)len && tab[a * stride] > e;
}

// src_bits (nullable, zeroed by the caller): the RAW-source words of the TLS
// guide, OR-ed in at the first writer of every raw read (see k_prof_count4)
template <int OP>
__global__ void __launch_bounds__(256) k_prof_classify(DLoop L, Tabs t, uint32_t *raw_bits, int64_t chunk,
                                                        int64_t *chunk_counts, int64_t *hdr, uint32_t *src_bits) {
  __shared__ unsigned long long s_cnt[3];
  __shared__ unsigned long long s_first;
  if (threadIdx.x < 3) s_cnt[threadIdx.x] = 0;
  if (threadIdx.x == 0) s_first = ~0ull;
  JP_CTA_SYNC();
  const int lane = threadIdx.x & 31;
  const int64_t warps = (int64_t)gridDim.x * (blockDim.x >> 5);
  unsigned long long c_raw = 0, c_war = 0, c_waw = 0, first = ~0ull;
  const int64_t tiles = (L.n + 31) >> 5;
  // PRIV_TMP: minR(T) == minW(T) (every T write is also its covered read)
  const int32_t *rT = OP == JP_OP_PRIV_TMP ? t.wT : t.rT;
  // each warp takes kUnroll consecutive tiles per step; all loads before any use
  for (int64_t tile0 = ((int64_t)blockIdx.x * (blockDim.x >> 5) + (threadIdx.x >> 5)) * kUnroll; tile0 < tiles;
       tile0 += warps * kUnroll) {
    int64_t ia[kUnroll], ib[kUnroll], ic[kUnroll];
#pragma unroll
    for (int u = 0; u < kUnroll; u++) {
      const int64_t i = ((tile0 + u) << 5) + lane;
      if (i < L.n) {
        if constexpr (OP == JP_OP_ADD_C) { ia[u] = ixl(L, L.w, i); ib[u] = ixl(L, L.r, i); }
        else if constexpr (OP == JP_OP_SAXPY) { ia[u] = ixl(L, L.w, i); }
        else if constexpr (OP == JP_OP_PRIV_TMP) { ia[u] = ixl(L, L.s, i); ib[u] = ixl(L, L.w, i); }
        else { ia[u] = ixl(L, L.w, i); ib[u] = ixl(L, L.r, i); ic[u] = ixl(L, L.r2, i); }
      }
    }
    bool raw[kUnroll], war[kUnroll], waw[kUnroll];
#pragma unroll
    for (int u = 0; u < kUnroll; u++) {   // table lookups, all issued before the ballots
      const int64_t i = ((tile0 + u) << 5) + lane;
      raw[u] = war[u] = waw[u] = false;
      if (i < L.n) {
        const int32_t e = enc_gid(L.base + i);
        auto src = [&](int64_t a) {   // mark the first writer of a raw read's address
          if (src_bits) {
            const int64_t jw = (int64_t)(0x7FFFFFFF - t.wA[(int64_t)a * t.as]) - L.base;
            atomicOr(&src_bits[jw >> 5], 1u << (jw & 31));
          }
        };
        if constexpr (OP == JP_OP_ADD_C) {
          war[u] = earlier(t.rA, ia[u], L.lenA, e, t.as);
          waw[u] = earlier(t.wA, ia[u], L.lenA, e, t.as);
          raw[u] = ib[u] == ia[u] ? waw[u] : earlier(t.wA, ib[u], L.lenA, e, t.as);   // r == w: one lookup
          if (raw[u]) src(ib[u]);
        } else if constexpr (OP == JP_OP_SAXPY) {
          raw[u] = earlier(t.wA, ia[u], L.lenA, e, t.as);
          war[u] = earlier(t.rA, ia[u], L.lenA, e, t.as);
          waw[u] = raw[u];   // the same address is the exposed read and the write
          if (raw[u]) src(ia[u]);
        } else if constexpr (OP == JP_OP_PRIV_TMP) {
          war[u] = earlier(rT, ia[u], L.lenT, e);
          waw[u] = earlier(t.wT, ia[u], L.lenT, e) || earlier(t.wA, ib[u], L.lenA, e, t.as);
        } else {
          war[u] = earlier(t.rA, ia[u], L.lenA, e, t.as);
          waw[u] = earlier(t.wA, ia[u], L.lenA, e, t.as);
          const bool r0 = ib[u] == ia[u] ? waw[u] : earlier(t.wA, ib[u], L.lenA, e, t.as);
          const bool r1 = ic[u] == ia[u] ? waw[u] : ic[u] == ib[u] ? r0 : earlier(t.wA, ic[u], L.lenA, e, t.as);
          raw[u] = r0 || r1;
          if (r0) src(ib[u]);
          if (r1) src(ic[u]);
        }
      }
    }
#pragma unroll
    for (int u = 0; u < kUnroll; u++) {
      const int64_t tile = tile0 + u;
      if (tile >= tiles) break;   // warp-uniform
      const unsigned bR = __ballot_sync(0xffffffffu, raw[u]);
      const unsigned bA = __ballot_sync(0xffffffffu, war[u]);
      const unsigned bW = __ballot_sync(0xffffffffu, waw[u]);
      if (lane == 0) {
        c_raw += __popc(bR); c_war += __popc(bA); c_waw += __popc(bW);
        if (raw_bits) raw_bits[tile] = bR;
        if (bR && first == ~0ull) first = (unsigned long long)(L.base + (tile << 5) + __ffs(bR) - 1);
        if (chunk_counts && (bR | bA | bW)) {
          int64_t c = (tile << 5) / chunk;
          if (bR) atomicAdd((unsigned long long *)&chunk_counts[3 * c + 0], (unsigned long long)__popc(bR));
          if (bA) atomicAdd((unsigned long long *)&chunk_counts[3 * c + 1], (unsigned long long)__popc(bA));
          if (bW) atomicAdd((unsigned long long *)&chunk_counts[3 * c + 2], (unsigned long long)__popc(bW));
        }
      }
    }
  }
  if (lane == 0) {
    if (c_raw) atomicAdd(&s_cnt[0], c_raw);
    if (c_war) atomicAdd(&s_cnt[1], c_war);
    if (c_waw) atomicAdd(&s_cnt[2], c_waw);
    if (first != ~0ull) atomicMin(&s_first, first);
  }
  JP_CTA_SYNC();
  if (threadIdx.x < 3 && s_cnt[threadIdx.x]) atomicAdd((unsigned long long *)&hdr[H_RAW + threadIdx.x], s_cnt[threadIdx.x]);
  if (threadIdx.x == 0 && s_first != ~0ull) atomicMin((unsigned long long *)&hdr[H_FIRST_RAW], s_first);
}

// ---------------------------------------------------------------------------
// TLS guide (profile-guided mode B).  Two bitmaps over
// local iterations, one bit per iteration, 32 iterations per word:
//   raw_i  some exposed read a of i has an earlier writer (minW table, pass 1);
//   src_j  the A-write of j is exposed-read by a later iteration (maxRx table).
// An in-window RAW violation needs a raw reader and a source writer (reading
// A7), so TLS windows stamp only source writes and check only raw reads: the
// same first violator, hence the same windows and statistics.
// Pass G1 fills maxRx[a] = latest gid with an exposed read of a (int32, empty
// -1): __match_any_sync groups the lanes of a warp that read the same address
// and only the group's highest lane (its latest iteration) issues the atomic.
template <int OP>
__global__ void __launch_bounds__(256) k_guide_maxr(DLoop L, int32_t *maxRx) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  const int64_t n_up = (L.n + 31) & ~(int64_t)31;   // whole warps for the match
  const int lane = threadIdx.x & 31;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n_up; i += stride) {
    const bool act = i < L.n;
    const int32_t g = (int32_t)(L.base + i);
    int32_t a0 = -1, a1 = -1;
    if (act) {
      if constexpr (OP == JP_OP_SAXPY) a0 = (int32_t)ixl(L, L.w, i);
      else if constexpr (OP == JP_OP_ADD_C) a0 = (int32_t)ixl(L, L.r, i);
      else if constexpr (OP == JP_OP_STENCIL2) { a0 = (int32_t)ixl(L, L.r, i); a1 = (int32_t)ixl(L, L.r2, i); }
    }
    if constexpr (OP != JP_OP_PRIV_TMP) {
      const unsigned grp = __match_any_sync(0xffffffffu, a0);
      if (act && (31 - __clz(grp)) == lane) atomicMax(&maxRx[a0], g);
      if constexpr (OP == JP_OP_STENCIL2) {
        const unsigned grp2 = __match_any_sync(0xffffffffu, a1);
        if (act && (31 - __clz(grp2)) == lane) atomicMax(&maxRx[a1], g);
      }
    }
  }
}

// Pass G2: the two bitmaps (ballot per warp tile).
template <int OP>
__global__ void __launch_bounds__(256) k_guide_bits(DLoop L, const int32_t *minW, const int32_t *maxRx,
                                                    uint32_t *raw_bits, uint32_t *src_bits) {
  const int lane = threadIdx.x & 31;
  const int64_t warps = (int64_t)gridDim.x * (blockDim.x >> 5);
  const int64_t tiles = (L.n + 31) >> 5;
  for (int64_t tile = (int64_t)blockIdx.x * (blockDim.x >> 5) + (threadIdx.x >> 5); tile < tiles; tile += warps) {
    const int64_t i = (tile << 5) + lane;
    bool raw = false, src = false;
    if (i < L.n && OP != JP_OP_PRIV_TMP) {
      const int64_t gid = L.base + i;
      const int32_t e = enc_gid(gid);
      const int64_t a = ixl(L, L.w, i);
      if constexpr (OP == JP_OP_SAXPY) raw = minW[a] > e;
      else raw = minW[ixl(L, L.r, i)] > e;
      if constexpr (OP == JP_OP_STENCIL2) raw = raw || minW[ixl(L, L.r2, i)] > e;
      src = maxRx[a] > (int32_t)gid;
    }
    const unsigned bR = __ballot_sync(0xffffffffu, raw), bS = __ballot_sync(0xffffffffu, src);
    if (lane == 0) { raw_bits[tile] = bR; src_bits[tile] = bS; }
  }
}

template <int OP>
__global__ void __launch_bounds__(256) k_validate(DLoop L, int64_t *hdr) {
  int64_t bad = 0;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < L.n; i += stride) {
    if constexpr (OP == JP_OP_ADD_C) {
      check(ixl(L, L.r, i), L.lenA, bad); check(ixl(L, L.w, i), L.lenA, bad);
    } else if constexpr (OP == JP_OP_SAXPY) {
      check(ixl(L, L.r, i), L.lenX, bad); check(ixl(L, L.w, i), L.lenA, bad);
    } else if constexpr (OP == JP_OP_PRIV_TMP) {
      check(ixl(L, L.r, i), L.lenX, bad); check(ixl(L, L.s, i), L.lenT, bad); check(ixl(L, L.w, i), L.lenA, bad);
    } else {
      check(ixl(L, L.r, i), L.lenA, bad); check(ixl(L, L.r2, i), L.lenA, bad); check(ixl(L, L.w, i), L.lenA, bad);
    }
  }
  for (int o = 16; o; o >>= 1) bad += __shfl_xor_sync(0xffffffffu, bad, o);
  if ((threadIdx.x & 31) == 0 && bad) atomicAdd((unsigned long long *)&hdr[H_BAD], (unsigned long long)bad);
}

// one index array against its length: 16-byte loads, four in flight per thread
// (a stream at HBM rate; the structural path's only pass before the run)
__global__ void __launch_bounds__(256) k_check_idx(const int32_t *p, int64_t n, int64_t len, int64_t *bad_out) {
  int64_t bad = 0;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x, tid = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  const int64_t head = ((uintptr_t)p & 15) ? (16 - ((uintptr_t)p & 15)) / 4 : 0;
  const int64_t h = head < n ? head : n;
  if (tid < h) bad += (uint32_t)p[tid] >= (uint64_t)len;
  const int4 *p4 = reinterpret_cast<const int4 *>(p + h);
  const int64_t nv = (n - h) >> 2;
  auto chk = [&](int4 v) {
    bad += ((uint32_t)v.x >= (uint64_t)len) + ((uint32_t)v.y >= (uint64_t)len) + ((uint32_t)v.z >= (uint64_t)len) +
           ((uint32_t)v.w >= (uint64_t)len);
  };
  int64_t v = tid;
  for (; v + 3 * stride < nv; v += 4 * stride) {
    const int4 a = __ldcs(p4 + v), b = __ldcs(p4 + v + stride), c = __ldcs(p4 + v + 2 * stride),
               d = __ldcs(p4 + v + 3 * stride);
    chk(a); chk(b); chk(c); chk(d);
  }
  for (; v < nv; v += stride) chk(__ldcs(p4 + v));
  for (int64_t i = h + 4 * nv + tid; i < n; i += stride) bad += (uint32_t)p[i] >= (uint64_t)len;
  for (int o = 16; o; o >>= 1) bad += __shfl_xor_sync(0xffffffffu, bad, o);
  if ((threadIdx.x & 31) == 0 && bad) atomicAdd((unsigned long long *)bad_out, (unsigned long long)bad);
}

static int grid_for(int64_t n, int threads, int per_sm) {
  int64_t need = (n + threads - 1) / threads;
  int64_t cap = (int64_t)num_sms() * per_sm;
  return (int)(need < 1 ? 1 : need < cap ? need : cap);
}
// grid-stride kernels with equal work per CTA: one wave of co-resident CTAs
// (a partial second wave at lower occupancy costs more than it hides)
static int grid_resident(const void *fn, int64_t n, int threads, size_t smem) {
  int per = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, fn, threads, smem) != cudaSuccess || per < 1) {
    cudaGetLastError();
    per = 4;
  }
  return grid_for(n, threads, per);
}

template <int OP, int DT>
static void run_stamp(const DLoop &d, Tabs t, int64_t *hdr, size_t smem, cudaStream_t st) {
  (void)DT;
  if (smem > 48 * 1024) cudaFuncSetAttribute(k_prof_stamp4<OP>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  const int64_t nq = (d.n + 3) / 4;
  k_prof_stamp4<OP><<<grid_resident((const void *)k_prof_stamp4<OP>, (nq + kQuadSteps - 1) / kQuadSteps, 256, smem), 256,
                      smem, st>>>(d, t, idx_vec(d), hdr);
  note_launch();
}

static Tabs tabs_of(const DLoop &d, void *ws, const Layout &lo) {
  Tabs t;
  t.lo = 0;
  t.span = 0xFFFFFFFFu;
  t.count_bad = 1;
  t.wA = at<int32_t>(ws, lo, R_MINW_A);
  t.rA = at<int32_t>(ws, lo, R_MINR_A);
  t.wT = at<int32_t>(ws, lo, R_MINW_T);
  t.rT = at<int32_t>(ws, lo, R_MINR_T);
  t.sA = t.wA && d.lenA <= kSmemSlots;
  t.sT = t.wT && d.lenT <= kSmemSlots;
  t.pA = nullptr;
  t.as = 1;
  return t;
}

// jp_schedule may stamp the A tables straight into interleaved {minW, minR}
// pairs held in the TLS write-log region (free until TLS, which resets it):
// large tables only (beyond L2), both tables present, region available
bool stamp_pairs_ok(const Job &j, void *ws, const Layout &lo) {
  const char *e = getenv("JP_CLASSIFY_PAIRS");
  if (e && e[0] == '0') return false;
  return lo.bytes[R_MINW_A] && lo.bytes[R_MINR_A] && lo.bytes[R_TLS_S_A] >= 8 * (size_t)j.d.lenA &&
         j.d.lenA >= (1 << 20) && j.d.lenA > kSmemSlots && j.op != JP_OP_PRIV_TMP &&
         (lo.off[R_TLS_S_A] & 15) == 0 && ws;
}

cudaError_t launch_prof_stamp(const Job &j, void *ws, const Layout &lo, cudaStream_t st, bool pairs, bool pairs_ready) {
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  cudaMemsetAsync(hdr, 0, kHeaderBytes, st);
  cudaMemsetAsync(&hdr[H_FIRST_RAW], 0xFF, sizeof(int64_t), st);   // none (= ~0 for the u64 atomicMin)
  size_t tab_bytes = 0;
  for (int r = R_MINW_A; r <= R_MINR_T; r++) {
    if (pairs && (r == R_MINW_A || r == R_MINR_A)) continue;
    if (lo.bytes[r]) cudaMemsetAsync(static_cast<char *>(ws) + lo.off[r], 0xFF, lo.bytes[r], st);
    tab_bytes += lo.bytes[r];
  }
  int32_t *pw = pairs ? at<int32_t>(ws, lo, R_TLS_S_A) : nullptr;
  if (pw) {
    if (!pairs_ready) cudaMemsetAsync(pw, 0xFF, 8 * (size_t)j.d.lenA, st);   // (else filled by the caller)
    tab_bytes += 8 * (size_t)j.d.lenA;
  }
  if (j.d.n == 0) return launch_check();
  Tabs t = tabs_of(j.d, ws, lo);
  if (pw) {
    t.wA = pw;
    t.rA = pw + 1;
    t.as = 2;
    t.sA = 0;
  }
  size_t smem = 0;
  if (t.sA) smem += (size_t)j.d.lenA * 4 * (t.rA ? 2 : 1);
  if (t.sT) smem += (size_t)j.d.lenT * 4;
  // tables beyond ~48 MB (a third of L2) are stamped one address window at a
  // time: every pass re-streams the index arrays but its random atomics hit L2
  const int64_t amax = std::max(j.d.lenA, j.d.lenT);
  const size_t pb = stamp_pass_bytes();
  int np = (t.sA || t.sT) ? 1 : (int)((tab_bytes + pb - 1) / pb);
  if (np < 1) np = 1;
  const int64_t step = (amax + np - 1) / np;
  for (int p = 0; p < np; p++) {
    t.lo = (uint32_t)(p * step);
    t.span = np == 1 ? 0xFFFFFFFFu : (uint32_t)step;
    t.count_bad = p == 0;
    JP_DISPATCH(j.op, j.dt, run_stamp, j.d, t, hdr, smem, st);
  }
  return launch_check();
}

__global__ void k_interleave(const int32_t *w, const int32_t *r, int2 *pairs, int64_t len);

template <int OP, int DT>
static void run_classify(const DLoop &d, Tabs t, uint32_t *bits, int64_t chunk, int64_t *cc, int64_t *hdr,
                         uint32_t *src_bits, cudaStream_t st) {
  (void)DT;
  int64_t tiles = (d.n + 31) / 32;
  if (!bits && !cc) {
    const int64_t nq = (d.n + 3) / 4;
    if constexpr (OP != JP_OP_PRIV_TMP) {
      if (t.pA) {   // large A tables: classify from interleaved {minW, minR} pairs
        if (t.as == 1)   // (not already stamped as pairs)
          k_interleave<<<grid_for(d.lenA / 4 + 1, 256, 8), 256, 0, st>>>(t.wA, t.rA, const_cast<int2 *>(t.pA), d.lenA);
        k_prof_count4<OP, false, true><<<grid_resident((const void *)k_prof_count4<OP, false, true>,
                                                       (nq + kQuadSteps - 1) / kQuadSteps, 256, 0), 256, 0, st>>>(
            d, t, idx_vec(d), hdr, nullptr, nullptr);
        note_launch(2);
        return;
      }
    }
    k_prof_count4<OP, false><<<grid_resident((const void *)k_prof_count4<OP, false>, (nq + kQuadSteps - 1) / kQuadSteps,
                                             256, 0), 256, 0, st>>>(d, t, idx_vec(d), hdr,
                                                                                                 nullptr, nullptr);
  } else if (cc && chunk >= 128 && (bits == nullptr) == (src_bits == nullptr) &&
             !(OP == JP_OP_PRIV_TMP && bits) && !getenv("JP_CLASSIFY_BALLOT")) {
    // chunk counts (and the guide words) from the quad kernel: 4 iterations per
    // lane, warp-aggregated chunk atomics (the stealing scheduler's profile)
    const int64_t nq = (d.n + 3) / 4;
    const int64_t g = (nq + kQuadSteps - 1) / kQuadSteps;
    if constexpr (OP != JP_OP_PRIV_TMP) {
      if (bits && t.pA) {
        k_prof_count4<OP, true, true><<<grid_resident((const void *)k_prof_count4<OP, true, true>, g, 256, 0), 256, 0,
                                        st>>>(d, t, idx_vec(d), hdr, bits, src_bits, chunk, cc);
      } else if (bits) {
        k_prof_count4<OP, true><<<grid_resident((const void *)k_prof_count4<OP, true>, g, 256, 0), 256, 0, st>>>(
            d, t, idx_vec(d), hdr, bits, src_bits, chunk, cc);
      } else if (t.pA) {   // stamped as pairs (no guide: restart recovery asked for)
        k_prof_count4<OP, false, true><<<grid_resident((const void *)k_prof_count4<OP, false, true>, g, 256, 0), 256,
                                         0, st>>>(d, t, idx_vec(d), hdr, nullptr, nullptr, chunk, cc);
      } else {
        k_prof_count4<OP, false><<<grid_resident((const void *)k_prof_count4<OP, false>, g, 256, 0), 256, 0, st>>>(
            d, t, idx_vec(d), hdr, nullptr, nullptr, chunk, cc);
      }
    } else {
      k_prof_count4<OP, false><<<grid_resident((const void *)k_prof_count4<OP, false>, g, 256, 0), 256, 0, st>>>(
          d, t, idx_vec(d), hdr, nullptr, nullptr, chunk, cc);
    }
  } else {
    k_prof_classify<OP><<<grid_resident((const void *)k_prof_classify<OP>, (tiles + kUnroll - 1) / kUnroll * 32, 256, 0),
                          256, 0, st>>>(d, t, bits, chunk, cc, hdr, src_bits);
  }
  note_launch();
}

// PRIV_TMP with identity Y writes and an indirect scratch index s: no exposed
// read of a written array (X is read-only, T's read is covered), so raw = 0,
// and war_i = waw_i = "an earlier iteration wrote T[s_i]" = "i is not the first
// writer of its slot".  Every slot whose (global) first writer lies in this
// range has exactly one such iteration, so war = waw = n - #{slots whose first
// writer is in [base, base + n)}: one pass over the small T table replaces the
// classify pass over the s stream.
__global__ void __launch_bounds__(1024) k_slot_first_writers(const int32_t *wT, int64_t lenT, int64_t base, int64_t n,
                                                             int64_t *hdr) {
  __shared__ unsigned long long cnt;
  if (threadIdx.x == 0) cnt = 0;
  __syncthreads();
  unsigned c = 0;
  for (int64_t a = threadIdx.x; a < lenT; a += blockDim.x) {
    const int32_t v = wT[a];
    if (v >= 0) {
      const int64_t gid = 0x7FFFFFFF - (int64_t)v;
      c += gid >= base && gid < base + n;
    }
  }
  c = __reduce_add_sync(0xffffffffu, c);
  if ((threadIdx.x & 31) == 0 && c) atomicAdd(&cnt, (unsigned long long)c);
  __syncthreads();
  if (threadIdx.x == 0) {
    hdr[H_RAW] = 0;
    hdr[H_WAR] = n - (int64_t)cnt;
    hdr[H_WAW] = n - (int64_t)cnt;
  }
}

static constexpr int64_t kSlotCountMaxT = 1 << 20;

cudaError_t launch_prof_classify(const Job &j, void *ws, const Layout &lo, uint32_t *raw_bits, int64_t chunk,
                                 int64_t *chunk_counts, cudaStream_t st, uint32_t *src_bits, bool stamped_pairs) {
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  cudaMemsetAsync(&hdr[H_RAW], 0, 3 * sizeof(int64_t), st);
  cudaMemsetAsync(&hdr[H_FIRST_RAW], 0xFF, sizeof(int64_t), st);
  if (chunk_counts) cudaMemsetAsync(chunk_counts, 0, sizeof(int64_t) * 3 * ((j.d.n + chunk - 1) / chunk), st);
  if (j.d.n == 0) return launch_check();
  Tabs t = tabs_of(j.d, ws, lo);
  // the one-CTA slot count reads all of T's table: taken only when that table is
  // small next to the s stream the full pass would read (config 4: 1024 slots)
  if (j.op == JP_OP_PRIV_TMP && !j.d.w && j.d.s && t.wT && !raw_bits && !chunk_counts && !src_bits &&
      j.d.lenT <= kSlotCountMaxT && j.d.lenT <= j.d.n / 8 + 1024 && !getenv("JP_CLASSIFY_FULL")) {
    k_slot_first_writers<<<1, 1024, 0, st>>>(t.wT, j.d.lenT, j.d.base, j.d.n, hdr);
    note_launch();
    return launch_check();
  }
  if (stamped_pairs) {   // the stamp pass wrote {minW, minR} pairs into region 7
    t.wA = at<int32_t>(ws, lo, R_TLS_S_A);
    t.rA = t.wA + 1;
    t.as = 2;
    t.pA = reinterpret_cast<const int2 *>(t.wA);
  }
  if (src_bits) cudaMemsetAsync(src_bits, 0, 4 * (size_t)((j.d.n + 31) / 32), st);
  // counts only, separate large A tables: interleave them into the TLS write-log
  // region (scratch until a TLS run resets it) and classify from the pairs
  unsigned long long *scratch = at<unsigned long long>(ws, lo, R_TLS_S_A);
  if (!stamped_pairs && !raw_bits && !chunk_counts && !src_bits && scratch && lo.bytes[R_TLS_S_A] >= 8 * (size_t)j.d.lenA &&
      t.wA && t.rA && !t.sA && j.d.lenA >= (1 << 20) && ((uintptr_t)t.wA & 15) == 0 && ((uintptr_t)t.rA & 15) == 0 &&
      getenv_int("JP_CLASSIFY_PAIRS", 1))
    t.pA = reinterpret_cast<const int2 *>(scratch);
  JP_DISPATCH(j.op, j.dt, run_classify, j.d, t, raw_bits, chunk, chunk_counts, hdr, src_bits, st);
  return launch_check();
}

// pairs[a] = {minW[a], minR[a]}: 16-byte loads of both tables, 16-byte stores
__global__ void __launch_bounds__(256) k_interleave(const int32_t *w, const int32_t *r, int2 *pairs, int64_t len) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x, nq = len >> 2;
  const int4 *w4 = reinterpret_cast<const int4 *>(w), *r4 = reinterpret_cast<const int4 *>(r);
  int4 *p4 = reinterpret_cast<int4 *>(pairs);
  for (int64_t q = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; q < nq; q += stride) {
    const int4 a = __ldcs(w4 + q), b = __ldcs(r4 + q);
    p4[2 * q] = make_int4(a.x, b.x, a.y, b.y);
    p4[2 * q + 1] = make_int4(a.z, b.z, a.w, b.w);
  }
  for (int64_t a = 4 * nq + (int64_t)blockIdx.x * blockDim.x + threadIdx.x; a < len; a += stride)
    pairs[a] = make_int2(w[a], r[a]);
}

template <int OP, int DT>
static void run_classify_guide(const DLoop &d, Tabs t, uint32_t *graw, uint32_t *gsrc, int64_t *hdr, cudaStream_t st) {
  (void)DT;
  const int64_t nq = (d.n + 3) / 4;
  const int g = grid_for((nq + kQuadSteps - 1) / kQuadSteps, 256, 8);
  auto *dist = reinterpret_cast<unsigned long long *>(hdr + H_DIST);
  if constexpr (OP == JP_OP_PRIV_TMP) {   // never guided: counts only
    k_prof_count4<OP, false><<<g, 256, 0, st>>>(d, t, idx_vec(d), hdr, nullptr, nullptr);
  } else {
    if (t.pA) {
      if (t.as == 1) {
        k_interleave<<<grid_for(d.lenA / 4 + 1, 256, 8), 256, 0, st>>>(t.wA, t.rA, const_cast<int2 *>(t.pA), d.lenA);
        note_launch();
      }
      k_prof_count4<OP, true, true><<<g, 256, 0, st>>>(d, t, idx_vec(d), hdr, graw, gsrc, 0, nullptr, dist);
    } else {
      k_prof_count4<OP, true><<<g, 256, 0, st>>>(d, t, idx_vec(d), hdr, graw, gsrc, 0, nullptr, dist);
    }
  }
  note_launch();
}

cudaError_t launch_prof_classify_guide(const Job &j, void *ws, const Layout &lo, cudaStream_t st, bool stamped_pairs) {
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  uint32_t *bits = at<uint32_t>(ws, lo, R_GUIDE);
  if (!bits) return launch_prof_classify(j, ws, lo, nullptr, 0, nullptr, st);
  cudaMemsetAsync(&hdr[H_RAW], 0, 3 * sizeof(int64_t), st);
  cudaMemsetAsync(&hdr[H_FIRST_RAW], 0xFF, sizeof(int64_t), st);
  cudaMemsetAsync(&hdr[H_DIST], 0, 32 * sizeof(int64_t), st);
  const int64_t nw = (j.d.n + 31) / 32;
  cudaMemsetAsync(bits + nw, 0, 4 * (size_t)nw, st);   // source words are OR-ed in
  if (j.d.n == 0) return launch_check();
  Tabs t = tabs_of(j.d, ws, lo);
  // the TLS write-log region (u64 [len_A], reset by every TLS launch) is free
  // until TLS runs: it holds the interleaved A tables for this pass when the
  // tables are large (beyond L2, where the second table's lookup is a DRAM burst)
  unsigned long long *scratch = at<unsigned long long>(ws, lo, R_TLS_S_A);
  if (stamped_pairs) {   // the stamp pass wrote the pairs: no interleave pass
    t.pA = reinterpret_cast<const int2 *>(scratch);
    t.wA = reinterpret_cast<int32_t *>(scratch);
    t.rA = t.wA + 1;
    t.as = 2;
  } else if (scratch && t.wA && t.rA && !t.sA && j.d.lenA >= (1 << 20) && ((uintptr_t)t.wA & 15) == 0 &&
             ((uintptr_t)t.rA & 15) == 0 && getenv_int("JP_CLASSIFY_PAIRS", 1)) {
    t.pA = reinterpret_cast<const int2 *>(scratch);
  }
  JP_DISPATCH(j.op, j.dt, run_classify_guide, j.d, t, bits, bits + nw, hdr, st);
  return launch_check();
}

template <int OP, int DT>
static void run_validate(const DLoop &d, int64_t *hdr, cudaStream_t st) {
  (void)DT;
  k_validate<OP><<<grid_for(d.n, 256, 8), 256, 0, st>>>(d, hdr);
  note_launch();
}

template <int OP, int DT>
static void run_guide(const DLoop &d, int32_t *minW, int32_t *maxRx, uint32_t *bits, cudaStream_t st) {
  (void)DT;
  const int64_t nw = (d.n + 31) / 32;
  k_guide_maxr<OP><<<grid_for(d.n, 256, 8), 256, 0, st>>>(d, maxRx);
  k_guide_bits<OP><<<grid_for(nw * 32, 256, 8), 256, 0, st>>>(d, minW, maxRx, bits, bits + nw);
  note_launch(2);
}

cudaError_t launch_tls_guide(const Job &j, void *ws, const Layout &lo, cudaStream_t st) {
  int32_t *maxRx = at<int32_t>(ws, lo, R_MAXRX_A);
  uint32_t *bits = at<uint32_t>(ws, lo, R_GUIDE);
  int32_t *minW = at<int32_t>(ws, lo, R_MINW_A);
  if (!bits || !maxRx || !minW || j.d.n == 0) return launch_check();
  cudaMemsetAsync(maxRx, 0xFF, lo.bytes[R_MAXRX_A], st);
  JP_DISPATCH(j.op, j.dt, run_guide, j.d, minW, maxRx, bits, st);
  return launch_check();
}

cudaError_t launch_validate_indirect(const Job &j, int64_t *bad, cudaStream_t st) {
  cudaMemsetAsync(bad, 0, sizeof(int64_t), st);
  const DLoop &d = j.d;
  auto one = [&](const int32_t *p, int64_t len) {
    if (!p || d.n == 0) return;
    k_check_idx<<<grid_for((d.n + 3) / 4, 256, 8), 256, 0, st>>>(p, d.n, len, bad);
    note_launch();
  };
  switch (j.op) {
    case JP_OP_ADD_C: one(d.r, d.lenA); one(d.w, d.lenA); break;
    case JP_OP_SAXPY: one(d.r, d.lenX); one(d.w, d.lenA); break;
    case JP_OP_PRIV_TMP: one(d.r, d.lenX); one(d.s, d.lenT); one(d.w, d.lenA); break;
    default: one(d.r, d.lenA); one(d.r2, d.lenA); one(d.w, d.lenA);
  }
  return launch_check();
}

cudaError_t launch_validate(const Job &j, int64_t *hdr, cudaStream_t st) {
  cudaMemsetAsync(&hdr[H_BAD], 0, sizeof(int64_t), st);
  if (j.d.n == 0) return launch_check();
  JP_DISPATCH(j.op, j.dt, run_validate, j.d, hdr, st);
  return launch_check();
}

}  // namespace jp

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
//   A1), then __ballot_sync + __popc per warp, one shared atomic per warp, one
//   global atomic per CTA; optional raw bitmap (D4) and per-chunk counts.
// The intra-warp / inter-warp split of the paper is an
// implementation detail here (reading A2): results do not depend on geometry.
#include "jp_host.h"

namespace jp {

struct Tabs {
  int32_t *wA, *rA, *wT, *rT;
  int sA, sT;   // pre-aggregate in shared memory
};

__device__ __forceinline__ void stamp(int32_t *g, int32_t *s, int64_t a, int64_t len, int32_t e, int64_t &bad) {
  if ((uint64_t)a >= (uint64_t)len) { bad++; return; }
  if (s) {
    if (s[a] < e) atomicMax(&s[a], e);
  } else if (g) {
    atomicMax(&g[a], e);
  }
}
__device__ __forceinline__ void check(int64_t a, int64_t len, int64_t &bad) {
  if ((uint64_t)a >= (uint64_t)len) bad++;
}

template <int OP>
__global__ void __launch_bounds__(256) k_prof_stamp(DLoop L, Tabs t, int64_t *hdr) {
  extern __shared__ int32_t sm[];
  int32_t *sAw = nullptr, *sAr = nullptr, *sTw = nullptr, *sTr = nullptr;
  int32_t *p = sm;
  if (t.sA) { sAw = p; p += L.lenA; if (t.rA) { sAr = p; p += L.lenA; } }
  if (t.sT) { sTw = p; p += L.lenT; sTr = p; p += L.lenT; }
  for (int64_t k = threadIdx.x; k < p - sm; k += blockDim.x) sm[k] = -1;
  JP_CTA_SYNC();

  int64_t bad = 0;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < L.n; i += stride) {
    const int32_t e = enc_gid(L.base + i);
    if constexpr (OP == JP_OP_ADD_C) {
      stamp(t.wA, sAw, ixl(L, L.w, i), L.lenA, e, bad);
      stamp(t.rA, sAr, ixl(L, L.r, i), L.lenA, e, bad);
    } else if constexpr (OP == JP_OP_SAXPY) {
      check(ixl(L, L.r, i), L.lenX, bad);
      int64_t a = ixl(L, L.w, i);
      stamp(t.wA, sAw, a, L.lenA, e, bad);
      if ((uint64_t)a < (uint64_t)L.lenA) stamp(t.rA, sAr, a, L.lenA, e, bad);
    } else if constexpr (OP == JP_OP_PRIV_TMP) {
      check(ixl(L, L.r, i), L.lenX, bad);
      int64_t a = ixl(L, L.s, i);
      stamp(t.wT, sTw, a, L.lenT, e, bad);
      if ((uint64_t)a < (uint64_t)L.lenT) stamp(t.rT, sTr, a, L.lenT, e, bad);
      stamp(t.wA, sAw, ixl(L, L.w, i), L.lenA, e, bad);
    } else {
      stamp(t.wA, sAw, ixl(L, L.w, i), L.lenA, e, bad);
      stamp(t.rA, sAr, ixl(L, L.r, i), L.lenA, e, bad);
      stamp(t.rA, sAr, ixl(L, L.r2, i), L.lenA, e, bad);
    }
  }
  // warp-aggregate the bad-index count
  for (int o = 16; o; o >>= 1) bad += __shfl_xor_sync(0xffffffffu, bad, o);
  if ((threadIdx.x & 31) == 0 && bad) atomicAdd((unsigned long long *)&hdr[H_BAD], (unsigned long long)bad);
  JP_CTA_SYNC();
  // flush the per-CTA pre-aggregated tables
  if (t.sA) {
    for (int64_t a = threadIdx.x; a < L.lenA; a += blockDim.x) {
      if (sAw[a] != -1) atomicMax(&t.wA[a], sAw[a]);
      if (sAr && sAr[a] != -1) atomicMax(&t.rA[a], sAr[a]);
    }
  }
  if (t.sT) {
    for (int64_t a = threadIdx.x; a < L.lenT; a += blockDim.x) {
      if (sTw[a] != -1) atomicMax(&t.wT[a], sTw[a]);
      if (sTr[a] != -1) atomicMax(&t.rT[a], sTr[a]);
    }
  }
}

// (bounds-guarded: classify may run before the host has seen the bad-index count)
__device__ __forceinline__ bool earlier(const int32_t *tab, int64_t a, int64_t len, int32_t e) {
  return tab && (uint64_t)a < (uint64_t)len && tab[a] > e;
}

template <int OP>
__global__ void __launch_bounds__(256) k_prof_classify(DLoop L, Tabs t, uint32_t *raw_bits, int64_t chunk,
                                                        int64_t *chunk_counts, int64_t *hdr) {
  __shared__ unsigned long long s_cnt[3];
  __shared__ unsigned long long s_first;
  if (threadIdx.x < 3) s_cnt[threadIdx.x] = 0;
  if (threadIdx.x == 0) s_first = ~0ull;
  JP_CTA_SYNC();
  const int lane = threadIdx.x & 31;
  const int64_t warps = (int64_t)gridDim.x * (blockDim.x >> 5);
  unsigned long long c_raw = 0, c_war = 0, c_waw = 0, first = ~0ull;
  const int64_t tiles = (L.n + 31) >> 5;
  for (int64_t tile = (int64_t)blockIdx.x * (blockDim.x >> 5) + (threadIdx.x >> 5); tile < tiles; tile += warps) {
    const int64_t i = (tile << 5) + lane;
    bool raw = false, war = false, waw = false;
    if (i < L.n) {
      const int32_t e = enc_gid(L.base + i);
      if constexpr (OP == JP_OP_ADD_C) {
        int64_t a = ixl(L, L.w, i);
        raw = earlier(t.wA, ixl(L, L.r, i), L.lenA, e);
        war = earlier(t.rA, a, L.lenA, e);
        waw = earlier(t.wA, a, L.lenA, e);
      } else if constexpr (OP == JP_OP_SAXPY) {
        int64_t a = ixl(L, L.w, i);
        raw = earlier(t.wA, a, L.lenA, e);
        war = earlier(t.rA, a, L.lenA, e);
        waw = raw;  // the same address is the exposed read and the write
      } else if constexpr (OP == JP_OP_PRIV_TMP) {
        int64_t a = ixl(L, L.s, i), b = ixl(L, L.w, i);
        war = earlier(t.rT, a, L.lenT, e);
        waw = earlier(t.wT, a, L.lenT, e) || earlier(t.wA, b, L.lenA, e);
      } else {
        int64_t a = ixl(L, L.w, i);
        raw = earlier(t.wA, ixl(L, L.r, i), L.lenA, e) || earlier(t.wA, ixl(L, L.r2, i), L.lenA, e);
        war = earlier(t.rA, a, L.lenA, e);
        waw = earlier(t.wA, a, L.lenA, e);
      }
    }
    const unsigned bR = __ballot_sync(0xffffffffu, raw);
    const unsigned bA = __ballot_sync(0xffffffffu, war);
    const unsigned bW = __ballot_sync(0xffffffffu, waw);
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

static int grid_for(int64_t n, int threads, int per_sm) {
  int64_t need = (n + threads - 1) / threads;
  int64_t cap = (int64_t)num_sms() * per_sm;
  return (int)(need < 1 ? 1 : need < cap ? need : cap);
}

template <int OP, int DT>
static void run_stamp(const DLoop &d, Tabs t, int64_t *hdr, size_t smem, cudaStream_t st) {
  (void)DT;
  if (smem > 48 * 1024) cudaFuncSetAttribute(k_prof_stamp<OP>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  k_prof_stamp<OP><<<grid_for(d.n, 256, 8), 256, smem, st>>>(d, t, hdr);
  note_launch();
}

static Tabs tabs_of(const DLoop &d, void *ws, const Layout &lo) {
  Tabs t;
  t.wA = at<int32_t>(ws, lo, R_MINW_A);
  t.rA = at<int32_t>(ws, lo, R_MINR_A);
  t.wT = at<int32_t>(ws, lo, R_MINW_T);
  t.rT = at<int32_t>(ws, lo, R_MINR_T);
  t.sA = t.wA && d.lenA <= kSmemSlots;
  t.sT = t.wT && d.lenT <= kSmemSlots;
  return t;
}

cudaError_t launch_prof_stamp(const Job &j, void *ws, const Layout &lo, cudaStream_t st) {
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  cudaMemsetAsync(hdr, 0, kHeaderBytes, st);
  cudaMemsetAsync(&hdr[H_FIRST_RAW], 0xFF, sizeof(int64_t), st);   // none (= ~0 for the u64 atomicMin)
  for (int r = R_MINW_A; r <= R_MINR_T; r++)
    if (lo.bytes[r]) cudaMemsetAsync(static_cast<char *>(ws) + lo.off[r], 0xFF, lo.bytes[r], st);
  if (j.d.n == 0) return launch_check();
  Tabs t = tabs_of(j.d, ws, lo);
  size_t smem = 0;
  if (t.sA) smem += (size_t)j.d.lenA * 4 * (t.rA ? 2 : 1);
  if (t.sT) smem += (size_t)j.d.lenT * 4 * 2;
  JP_DISPATCH(j.op, j.dt, run_stamp, j.d, t, hdr, smem, st);
  return launch_check();
}

template <int OP, int DT>
static void run_classify(const DLoop &d, Tabs t, uint32_t *bits, int64_t chunk, int64_t *cc, int64_t *hdr,
                         cudaStream_t st) {
  (void)DT;
  int64_t tiles = (d.n + 31) / 32;
  k_prof_classify<OP><<<grid_for(tiles * 32, 256, 8), 256, 0, st>>>(d, t, bits, chunk, cc, hdr);
  note_launch();
}

cudaError_t launch_prof_classify(const Job &j, void *ws, const Layout &lo, uint32_t *raw_bits, int64_t chunk,
                                 int64_t *chunk_counts, cudaStream_t st) {
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  cudaMemsetAsync(&hdr[H_RAW], 0, 3 * sizeof(int64_t), st);
  cudaMemsetAsync(&hdr[H_FIRST_RAW], 0xFF, sizeof(int64_t), st);
  if (chunk_counts) cudaMemsetAsync(chunk_counts, 0, sizeof(int64_t) * 3 * ((j.d.n + chunk - 1) / chunk), st);
  if (j.d.n == 0) return launch_check();
  Tabs t = tabs_of(j.d, ws, lo);
  JP_DISPATCH(j.op, j.dt, run_classify, j.d, t, raw_bits, chunk, chunk_counts, hdr, st);
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

cudaError_t launch_validate(const Job &j, int64_t *hdr, cudaStream_t st) {
  cudaMemsetAsync(&hdr[H_BAD], 0, sizeof(int64_t), st);
  if (j.d.n == 0) return launch_check();
  JP_DISPATCH(j.op, j.dt, run_validate, j.d, hdr, st);
  return launch_check();
}

}  // namespace jp

// jp_bucket.cu -- the dependency-density profile of a loop over a large A by
// address buckets (P1 stamp + P2 classify of SURVEY Sec.8(a); the paper's
// profiler, Fig. 1 "DD analysis"; densities per reading A1).
//
// The two-pass stamp/classify profile (jp_profile.cu) needs one random L2 atomic
// per access (first writer / first reader of the address) and then random reads
// of the same tables: on config 3 (N = len_A = 2^24) that is 2^25 atomics at the
// L2 atomic rate (3 address-window passes) plus a classify pass whose lookups
// miss L2 -- 1.6 GB of DRAM traffic for 0.47 GB of algorithmic bytes.  Here the
// accesses are first PARTITIONED by address instead, so every first-writer /
// first-reader table lives in one CTA's shared memory:
//
//   count    per tile of 16384 iterations: accesses per bucket of 8192
//            addresses (shared-memory histogram), and the out-of-range count;
//   scan     per bucket, the tiles' exclusive offsets; then the buckets' bases;
//   scatter  every access as an 8-byte record (iteration, address in its
//            bucket, write / read) into its bucket's segment, tile by tile:
//            staged in shared memory grouped by bucket first, so each (tile,
//            bucket) run is written as one contiguous piece (random 4-byte
//            stores were bound by L2 transactions: 345 us on config 3);
//   evaluate one CTA per bucket: minW / minR of its 8192 addresses by shared
//            atomics over the bucket's records, then every record evaluated
//            against them -- raw (an exposed read whose first writer is
//            earlier), war / waw (a write whose first reader / writer is
//            earlier) -- with the per-iteration guide bits, the RAW-source bits
//            (the first writer of every raw read), the raw-distance histogram,
//            the first raw iteration and optional per-chunk counts.
//
// DRAM traffic per iteration (ADD_C): index streams twice (16 B), records
// written and read once (2 x 2 x 8 B); the tables never leave shared memory.
// (4-byte records holding the iteration within its tile were measured slower:
// recovering the tile of every record costs more instructions than the bytes.)
// Counts are per access: ADD_C has exactly one write and one exposed read of A
// per iteration (raw from the read, war / waw from the write); SAXPY's only A
// access is Y[w], read and written by the same iteration, so raw = war = waw =
// "an earlier iteration wrote this address" (one write record).
#include <algorithm>
#include <string>
#include <vector>
#include "jp_host.h"

namespace jp {

constexpr int kBShift = 13;                 // addresses per bucket: 8192
constexpr int kBSpan = 1 << kBShift;
constexpr int kTShift = 14;                 // iterations per tile: 16384
constexpr int kTile = 1 << kTShift;
constexpr int kBThreads = 1024;
constexpr int kEvalThreads = 512;
constexpr int kMaxBuckets = 8192;           // len_A <= 2^26
constexpr int kMaxTiles = 16384;            // n <= 2^26
constexpr int kSmemChunks = 1024;           // per-chunk counts kept in shared memory up to this many chunks
// record (8 bytes): local iteration (low word) | address in the bucket << 32 | write << 63
// | also-read << 62: an ADD_C iteration whose read and write are the same address
// (an in-place update, A[w[i]] = A[w[i]] + c) files ONE record for both accesses
constexpr unsigned long long kRecW = 1ull << 63, kRecRW = 1ull << 62;
__device__ __forceinline__ bool rec_reads(unsigned long long x) { return !(x & kRecW) || (x & kRecRW); }

struct BkView {
  const int32_t *r, *w;   // ADD_C: read r, write w; SAXPY: w only (NULL => identity ioff + i)
  int64_t n, ioff;
  uint32_t lenA;
  int B, T;
  uint32_t *crange;       // nullable: per chunk min / max address (chunk = ctiles tiles)
  int ctiles;
  const int64_t *gate;    // nullable: the header's H_GATE word -- every kernel exits when it is nonzero
};
__device__ __forceinline__ bool gated(const int64_t *g) { return g && *(volatile const int64_t *)g != 0; }

__device__ __forceinline__ int4 ld_idx4(const int32_t *p, int64_t i, int64_t n, int64_t ioff, bool vec) {
  if (!p) {
    const int b = (int)(ioff + i);
    return make_int4(b, b + 1, b + 2, b + 3);
  }
  if (vec && i + 4 <= n) return __ldcs(reinterpret_cast<const int4 *>(p + i));
  int4 v;
  v.x = p[i];
  v.y = i + 1 < n ? p[i + 1] : 0;
  v.z = i + 2 < n ? p[i + 2] : 0;
  v.w = i + 3 < n ? p[i + 3] : 0;
  return v;
}
__device__ __forceinline__ int q4(const int4 &v, int k) { return k == 0 ? v.x : k == 1 ? v.y : k == 2 ? v.z : v.w; }

// Visit the accesses of tile blockIdx.x four iterations at a time (16-byte
// index loads, kU quads in flight per lane): f(a[8], wr[8], il0, kn) gets the
// quad's accesses -- ADD_C: (w, r) of each of the kn <= 4 iterations, SAXPY: w.
template <int OP, int kU = 4, typename F>
__device__ __forceinline__ void for_tile(const BkView &V, bool vec, F &&f) {
  const int64_t t0 = (int64_t)blockIdx.x << kTShift;
  const int64_t tn = V.n - t0 < kTile ? V.n - t0 : kTile;
  const int nq = (int)((tn + 3) >> 2);
  for (int q0 = threadIdx.x; q0 < nq; q0 += kBThreads * kU) {
    int4 vw[kU], vr[kU];
#pragma unroll
    for (int u = 0; u < kU; u++) {
      const int q = q0 + u * kBThreads;
      if (q < nq) {
        vw[u] = ld_idx4(V.w, t0 + 4 * q, V.n, V.ioff, vec);
        if constexpr (OP == JP_OP_ADD_C) vr[u] = ld_idx4(V.r, t0 + 4 * q, V.n, V.ioff, vec);
      }
    }
#pragma unroll
    for (int u = 0; u < kU; u++) {
      const int q = q0 + u * kBThreads;
      if (q >= nq) break;
      const int kn = tn - 4 * q < 4 ? (int)(tn - 4 * q) : 4;
      f(vw[u], vr[u], 4 * q, kn);
    }
  }
}

// cnt[t * B + b] = records of tile t in bucket b: writes (an also-read record
// included) in the low 16 bits, pure reads << 16 (a tile holds at most 16384 of
// each); out-of-range indices counted into *bad
template <int OP>
__global__ void __launch_bounds__(kBThreads, 2) k_bk_count(BkView V, int vec, uint32_t *cnt, int64_t *bad) {
  if (gated(V.gate)) return;
  extern __shared__ uint32_t h[];
  for (int b = threadIdx.x; b < V.B; b += kBThreads) h[b] = 0;
  __syncthreads();
  unsigned nbad = 0;
  uint32_t mn = 0xFFFFFFFFu, mx = 0u;   // the tile's address range (crange: a tile lies in one chunk)
  // an out-of-range index is counted (the profile then fails) and filed under
  // bucket 0, consistently with the scatter below
  // (two quads in flight per lane: 32 registers, two CTAs per SM)
  for_tile<OP, 2>(V, vec, [&](const int4 &w4, const int4 &r4, int, int kn) {
#pragma unroll
    for (int k = 0; k < 4; k++) {
      if (k < kn) {
        const uint32_t a = (uint32_t)q4(w4, k);
        const bool oka = a < V.lenA;
        nbad += !oka;
        atomicAdd(&h[oka ? a >> kBShift : 0], 1u);
        if (oka) { mn = min(mn, a); mx = max(mx, a); }
        if constexpr (OP == JP_OP_ADD_C) {
          const uint32_t c = (uint32_t)q4(r4, k);
          const bool okc = c < V.lenA;
          nbad += !okc;
          if (c != a) atomicAdd(&h[okc ? c >> kBShift : 0], 1u << 16);   // (c == a: one record for both)
          if (okc) { mn = min(mn, c); mx = max(mx, c); }
        }
      }
    }
  });
  nbad = __reduce_add_sync(0xffffffffu, nbad);
  if ((threadIdx.x & 31) == 0 && nbad) atomicAdd(reinterpret_cast<unsigned long long *>(bad), (unsigned long long)nbad);
  if (V.crange) {
    mn = __reduce_min_sync(0xffffffffu, mn);
    mx = __reduce_max_sync(0xffffffffu, mx);
    if ((threadIdx.x & 31) == 0 && mn <= mx) {
      const int c = blockIdx.x / V.ctiles;
      atomicMin(&V.crange[2 * c], mn);
      atomicMax(&V.crange[2 * c + 1], mx);
    }
  }
  __syncthreads();
  uint32_t *row = cnt + (size_t)blockIdx.x * V.B;
  for (int b = threadIdx.x; b < V.B; b += kBThreads) row[b] = h[b];
}

// per bucket: exclusive prefix over the tiles (in place) of the records kept and
// the bucket total.  A bucket no iteration writes drops its pure reads (a read
// with no writer of its address is neither raw nor the first read of a written
// address: it changes no count, guide bit or table of the profile): wflag[b].
// Block = 16 buckets x 64 tile segments (two segments per warp).
constexpr int kScanNB = 16, kScanNS = 1024 / kScanNB;   // buckets x tile segments per CTA (B / 16 CTAs)
__global__ void __launch_bounds__(1024) k_bk_scan_tiles(uint32_t *cnt, int T, int B, uint32_t *tot,
                                                         uint32_t *wflag, const int64_t *gate) {
  if (gated(gate)) return;
  __shared__ uint32_t part_w[kScanNS][kScanNB + 1], part_r[kScanNS][kScanNB + 1];
  const int lane = threadIdx.x % kScanNB, seg = threadIdx.x / kScanNB;
  const int b = blockIdx.x * kScanNB + lane;
  const int per = (T + kScanNS - 1) / kScanNS, t0 = seg * per, t1 = min(T, t0 + per);
  uint32_t sw = 0, sr = 0;
  if (b < B)
#pragma unroll 8
    for (int t = t0; t < t1; t++) {
      const uint32_t c = cnt[(size_t)t * B + b];
      sw += c & 0xFFFFu;
      sr += c >> 16;
    }
  part_w[seg][lane] = sw;
  part_r[seg][lane] = sr;
  __syncthreads();
  uint32_t allw = 0;
  for (int k = 0; k < kScanNS; k++) allw += part_w[k][lane];
  const bool keep = allw > 0;
  uint32_t run = 0;
  for (int k = 0; k < seg; k++) run += part_w[k][lane] + (keep ? part_r[k][lane] : 0u);
  if (b < B) {
#pragma unroll 8
    for (int t = t0; t < t1; t++) {
      const uint32_t c = cnt[(size_t)t * B + b];
      cnt[(size_t)t * B + b] = run;
      run += (c & 0xFFFFu) + (keep ? c >> 16 : 0u);
    }
    if (seg == kScanNS - 1) {
      tot[b] = run;
      wflag[b] = keep ? 1u : 0u;
    }
  }
}

// base[b] = exclusive prefix of tot over the buckets (one CTA)
// ... and order[]: the buckets by decreasing record count (binned by floor log2),
// the order the one-CTA-per-bucket passes take them in, so that a few heavy
// buckets do not form the last wave (config 5: its WAW tail's buckets hold 3x
// the records of the others)
__global__ void __launch_bounds__(1024) k_bk_scan_buckets(const uint32_t *tot, int B, uint32_t *base,
                                                           uint32_t *order, const int64_t *gate) {
  if (gated(gate)) return;
  __shared__ uint32_t ws[32];
  __shared__ uint32_t bin[33];
  const int per = (B + 1023) / 1024, b0 = threadIdx.x * per;
  uint32_t s = 0;
  for (int k = 0; k < per && b0 + k < B; k++) s += tot[b0 + k];
  uint32_t x = s;   // inclusive warp scan
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
    if ((threadIdx.x & 31) >= o) x += y;
  }
  if ((threadIdx.x & 31) == 31) ws[threadIdx.x >> 5] = x;
  __syncthreads();
  if (threadIdx.x < 32) {
    uint32_t v = ws[threadIdx.x];
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, v, o);
      if (threadIdx.x >= o) v += y;
    }
    ws[threadIdx.x] = v;
  }
  __syncthreads();
  uint32_t run = x - s + ((threadIdx.x >> 5) ? ws[(threadIdx.x >> 5) - 1] : 0);
  for (int k = 0; k < per && b0 + k < B; k++) {
    base[b0 + k] = run;
    run += tot[b0 + k];
  }
  if (!order) return;
  if (threadIdx.x < 33) bin[threadIdx.x] = 0;
  __syncthreads();
  for (int k = 0; k < per && b0 + k < B; k++) atomicAdd(&bin[32 - __clz(tot[b0 + k])], 1u);   // 0..32
  __syncthreads();
  if (threadIdx.x == 0) {   // exclusive starts, heaviest bin first
    uint32_t r = 0;
    for (int q = 32; q >= 0; q--) { const uint32_t c = bin[q]; bin[q] = r; r += c; }
  }
  __syncthreads();
  for (int k = 0; k < per && b0 + k < B; k++) order[atomicAdd(&bin[32 - __clz(tot[b0 + k])], 1u)] = (uint32_t)(b0 + k);
}

// records, tile-ordered inside each bucket's segment.  Shared memory: the
// tile's records staged by bucket (2 x 16384 x 4 B), the local bucket starts
// and cursors (B each), the global start of this tile's run in every bucket.
template <int OP>
__global__ void __launch_bounds__(kBThreads) k_bk_scatter(BkView V, int vec, const uint32_t *off, const uint32_t *tot,
                                                         const uint32_t *base, const uint32_t *wflag,
                                                         unsigned long long *rec) {
  if (gated(V.gate)) return;
  // staging: 6 bytes per record -- il | address in the bucket << 14 | write << 31,
  // and the bucket (16 bits) -- so that a 16384-iteration tile fits one SM
  extern __shared__ uint32_t sm32[];
  uint32_t *stage = sm32;                                      // [2 * kTile]
  uint16_t *stb = reinterpret_cast<uint16_t *>(stage + 2 * kTile);      // [2 * kTile]
  uint32_t *lpos = reinterpret_cast<uint32_t *>(stb + 2 * kTile);       // [B + 1] local exclusive starts
  uint32_t *cur = lpos + V.B + 1;                              // [B]
  uint32_t *gpos = cur + V.B;                                  // [B] global start of this tile's run
  uint8_t *wf = reinterpret_cast<uint8_t *>(gpos + V.B);       // [B] the bucket is written (else drop pure reads)
  __shared__ uint32_t wsum[kBThreads / 32];
  const int t = blockIdx.x, B = V.B;
  const uint32_t i0 = (uint32_t)t << kTShift;
  const uint32_t *row = off + (size_t)t * B, *nxt = t + 1 < V.T ? row + B : nullptr;
  // local counts -> exclusive scan over the buckets (per thread a contiguous run)
  const int per = (B + kBThreads - 1) / kBThreads, b0 = threadIdx.x * per;
  uint32_t s = 0;
  for (int k = 0; k < per && b0 + k < B; k++) {
    const int b = b0 + k;
    const uint32_t c = (nxt ? nxt[b] : tot[b]) - row[b];
    cur[b] = c;   // (count, for the scan below)
    gpos[b] = base[b] + row[b];
    wf[b] = (uint8_t)wflag[b];
    s += c;
  }
  uint32_t x = s;
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
    if ((threadIdx.x & 31) >= o) x += y;
  }
  if ((threadIdx.x & 31) == 31) wsum[threadIdx.x >> 5] = x;
  __syncthreads();
  uint32_t wpre = 0;
  for (int k = 0; k < (int)(threadIdx.x >> 5); k++) wpre += wsum[k];
  uint32_t run = wpre + x - s;
  for (int k = 0; k < per && b0 + k < B; k++) {
    const int b = b0 + k;
    const uint32_t c = cur[b];
    lpos[b] = run;
    cur[b] = run;
    run += c;
  }
  if (threadIdx.x == kBThreads - 1) lpos[B] = run;
  __syncthreads();
  for_tile<OP>(V, vec, [&](const int4 &w4, const int4 &r4, int il0, int kn) {
    // all positions of the quad first (the shared atomics issue back to back),
    // then the staging stores
    constexpr int kA = OP == JP_OP_ADD_C ? 8 : 4;
    uint32_t a[kA], pos[kA];
#pragma unroll
    for (int k = 0; k < 4; k++) {
      a[OP == JP_OP_ADD_C ? 2 * k : k] = (uint32_t)q4(w4, k);
      if constexpr (OP == JP_OP_ADD_C) a[2 * k + 1] = (uint32_t)q4(r4, k);
    }
    // an iteration reading the address it writes: one record (write | also-read)
    bool same[4];
#pragma unroll
    for (int k = 0; k < 4; k++) same[k] = OP == JP_OP_ADD_C && a[2 * k] == a[2 * k + 1];
    // skip[m]: a read folded into its iteration's write record, or a pure read of
    // a bucket nobody writes (dropped, see k_bk_scan_tiles)
    bool skip[kA];
#pragma unroll
    for (int m = 0; m < kA; m++) {
      if (a[m] >= V.lenA) a[m] = 0;   // (the count pass filed it under bucket 0 too)
      const int k = OP == JP_OP_ADD_C ? m >> 1 : m;
      skip[m] = OP == JP_OP_ADD_C && (m & 1) && (same[k] || !wf[a[m] >> kBShift]);
      pos[m] = k < kn && !skip[m] ? atomicAdd(&cur[a[m] >> kBShift], 1u) : 0u;
    }
#pragma unroll
    for (int m = 0; m < kA; m++) {
      const int k = OP == JP_OP_ADD_C ? m >> 1 : m;
      const bool wr = OP == JP_OP_ADD_C ? (m & 1) == 0 : true;
      if (k < kn && !skip[m]) {
        stage[pos[m]] = (uint32_t)(il0 + k) | (a[m] & (kBSpan - 1)) << kTShift | (wr ? 1u << 31 : 0u) |
                        (wr && same[k] ? 1u << 30 : 0u);
        stb[pos[m]] = (uint16_t)(a[m] >> kBShift);
      }
    }
  });
  __syncthreads();
  // copy out, flat: staged record k of bucket b goes to k + (gpos[b] - lpos[b])
  // (consecutive k of one run are consecutive records of the bucket's segment)
  for (int b = threadIdx.x; b < B; b += kBThreads) gpos[b] -= lpos[b];
  __syncthreads();
  const uint32_t nrec = lpos[B];
  for (uint32_t k = threadIdx.x; k < nrec; k += kBThreads) {
    const uint32_t x = stage[k];
    rec[k + gpos[stb[k]]] = (unsigned long long)(i0 + (x & (kTile - 1))) |
                            (unsigned long long)((x >> kTShift) & (kBSpan - 1)) << 32 | (x >> 31 ? kRecW : 0ull) |
                            ((x >> 30) & 1u ? kRecRW : 0ull);
  }
}

struct BkOut {
  int64_t *hdr;               // H_RAW / H_WAR / H_WAW, H_FIRST_RAW, H_DIST
  uint32_t *graw, *gsrc;      // guide words (nullable), zeroed by the caller
  int64_t chunk;              // per-chunk counts (cc nullable)
  int64_t *cc;
  int64_t gbase;              // global id of local iteration 0
  int32_t *wsrc;              // nullable: wsrc[i] = the first writer of raw iteration i's read (ADD_C)
  const uint32_t *order;      // nullable: bucket of CTA k (heaviest first)
  unsigned long long *vclr;   // nullable: V[a] = 0 at every raw read's address (the one-window TLS
                              // shadow slots a violator polls: no full clear of V needed)
};

template <int OP>
__global__ void __launch_bounds__(kEvalThreads) k_bk_eval(BkView V, const uint32_t *base, const uint32_t *tot,
                                                          const unsigned long long *rec, BkOut O) {
  if (gated(V.gate)) return;
  // dynamic: minW[8192], minR[8192] (ADD_C), then 3 x nch per-chunk counts when they fit
  extern __shared__ uint32_t s_dyn[];
  uint32_t *minW = s_dyn;
  uint32_t *minR = s_dyn + kBSpan;
  uint32_t *s_cc = s_dyn + (OP == JP_OP_ADD_C ? 2 : 1) * kBSpan;
  __shared__ unsigned s_dist[32];
  __shared__ unsigned long long s_cnt[3], s_first;
  const int b = O.order ? (int)O.order[blockIdx.x] : (int)blockIdx.x;
  const int nch = O.cc ? (int)((V.n + O.chunk - 1) / O.chunk) : 0;
  const bool cc_smem = O.cc && nch <= kSmemChunks;
  for (int k = threadIdx.x; k < kBSpan; k += kEvalThreads) {
    minW[k] = 0xFFFFFFFFu;
    if constexpr (OP == JP_OP_ADD_C) minR[k] = 0xFFFFFFFFu;
  }
  const uint32_t total = tot[b];
  if (threadIdx.x < 32) s_dist[threadIdx.x] = 0;
  if (threadIdx.x < 3) s_cnt[threadIdx.x] = 0;
  if (threadIdx.x == 0) s_first = ~0ull;
  if (cc_smem)
    for (int k = threadIdx.x; k < 3 * nch; k += kEvalThreads) s_cc[k] = 0;
  __syncthreads();
  const unsigned long long *rb = rec + base[b];
  constexpr int kU = 4;   // records in flight per thread
  auto sweep = [&](auto &&f) {
    for (uint32_t p0 = threadIdx.x; p0 < total; p0 += kEvalThreads * kU) {
      unsigned long long xv[kU];
#pragma unroll
      for (int u = 0; u < kU; u++) {
        const uint32_t p = p0 + (uint32_t)u * kEvalThreads;
        xv[u] = p < total ? rb[p] : 0ull;
      }
#pragma unroll
      for (int u = 0; u < kU; u++)
        if (p0 + (uint32_t)u * kEvalThreads < total) f(xv[u]);
    }
  };
  // pass 1: first writer / first reader of every address of the bucket
  sweep([&](unsigned long long x) {
    const uint32_t i = (uint32_t)x, al = (uint32_t)(x >> 32) & (kBSpan - 1);
    if (x & kRecW) atomicMin(&minW[al], i);
    if constexpr (OP == JP_OP_ADD_C)
      if (rec_reads(x)) atomicMin(&minR[al], i);
  });
  __syncthreads();
  // pass 2: every access against the final tables
  unsigned c_raw = 0, c_war = 0, c_waw = 0;
  unsigned long long first = ~0ull;
  sweep([&](unsigned long long x) {
    const uint32_t i = (uint32_t)x, al = (uint32_t)(x >> 32) & (kBSpan - 1);
    const uint32_t jw = minW[al];
    bool raw, war = false, waw = false;
    if (x & kRecW) {
      waw = jw < i;
      war = (OP == JP_OP_ADD_C ? minR[al] : jw) < i;   // (an also-read record's own read is minR = i: not < i)
      raw = OP == JP_OP_SAXPY ? waw : (x & kRecRW) && waw;
    } else {
      raw = jw < i;
    }
    c_raw += raw; c_war += war; c_waw += waw;
    if (raw) {
      if (O.wsrc && rec_reads(x)) O.wsrc[i] = (int32_t)jw;
      if (O.vclr && rec_reads(x)) O.vclr[(uint32_t)b << kBShift | al] = 0ull;
      if (O.graw) atomicOr(&O.graw[i >> 5], 1u << (i & 31));
      if (O.gsrc) atomicOr(&O.gsrc[jw >> 5], 1u << (jw & 31));
      atomicAdd(&s_dist[31 - __clz(i - jw)], 1u);
      if ((unsigned long long)i < first) first = i;
    }
    if (O.cc && (raw | war | waw)) {
      const int64_t ch = (int64_t)i / O.chunk;
      if (cc_smem) {
        if (raw) atomicAdd(&s_cc[3 * ch + 0], 1u);
        if (war) atomicAdd(&s_cc[3 * ch + 1], 1u);
        if (waw) atomicAdd(&s_cc[3 * ch + 2], 1u);
      } else {
        if (raw) atomicAdd(reinterpret_cast<unsigned long long *>(&O.cc[3 * ch + 0]), 1ull);
        if (war) atomicAdd(reinterpret_cast<unsigned long long *>(&O.cc[3 * ch + 1]), 1ull);
        if (waw) atomicAdd(reinterpret_cast<unsigned long long *>(&O.cc[3 * ch + 2]), 1ull);
      }
    }
  });
  c_raw = __reduce_add_sync(0xffffffffu, c_raw);
  c_war = __reduce_add_sync(0xffffffffu, c_war);
  c_waw = __reduce_add_sync(0xffffffffu, c_waw);
  for (int o = 16; o; o >>= 1) {
    const unsigned long long y = __shfl_xor_sync(0xffffffffu, first, o);
    first = y < first ? y : first;
  }
  if ((threadIdx.x & 31) == 0) {
    if (c_raw) atomicAdd(&s_cnt[0], (unsigned long long)c_raw);
    if (c_war) atomicAdd(&s_cnt[1], (unsigned long long)c_war);
    if (c_waw) atomicAdd(&s_cnt[2], (unsigned long long)c_waw);
    if (first != ~0ull) atomicMin(&s_first, first);
  }
  __syncthreads();
  if (threadIdx.x < 3 && s_cnt[threadIdx.x])
    atomicAdd(reinterpret_cast<unsigned long long *>(&O.hdr[H_RAW + threadIdx.x]), s_cnt[threadIdx.x]);
  if (threadIdx.x == 0 && s_first != ~0ull)
    atomicMin(reinterpret_cast<unsigned long long *>(&O.hdr[H_FIRST_RAW]), (unsigned long long)O.gbase + s_first);
  if (threadIdx.x < 32 && s_dist[threadIdx.x])
    atomicAdd(reinterpret_cast<unsigned long long *>(&O.hdr[H_DIST + threadIdx.x]), (unsigned long long)s_dist[threadIdx.x]);
  if (cc_smem)
    for (int k = threadIdx.x; k < 3 * nch; k += kEvalThreads)
      if (s_cc[k]) atomicAdd(reinterpret_cast<unsigned long long *>(&O.cc[k]), (unsigned long long)s_cc[k]);
}

// ---------------------------------------------------------------------------
// The last earlier writer of every raw read (reading B14, path 9).  With WAW a
// raw read of address a at iteration i must see the value of
// pred(i) = max{ j < i : w[j] = a } (the sequential semantics);
// the first-writer tables above do not hold it.  One CTA per bucket, over the
// records the profile left in place:
//   count    writers per address (shared atomics);
//   scan     the address segments of a writer list;
//   fill     every writer's iteration into its address's segment (unordered);
//   reads    pred(i) = the largest listed writer below i -> pred[i], and the
//            writer's publish bit; a read with no earlier writer of an address
//            that IS written (an exposed read, WAR on the window-start value)
//            marks the address;
//   writers  per address, its last writer: commit at once (now) or, when the
//            address has an exposed read, after the flow kernel's barrier (later).
// A bucket whose writers do not fit shared memory, or an address with more than
// kPredSegCap writers, fails the pass (H_PRED_FAIL): the caller keeps the
// windowed paths.  ADD_C only (one exposed read, one write per iteration).
// ---------------------------------------------------------------------------
// Two tiers: 512-thread CTAs, two per SM, hold up to kPredCapS writers per bucket;
// a bucket with more is marked and redone by the second launch (1024 threads,
// one CTA per SM, the whole 226 KB), which skips every other bucket.
constexpr uint32_t kPredSegCap = 4096;
constexpr size_t kPredSmemS = 110 * 1024, kPredSmemB = 226 * 1024;   // (+ static <= the 227 KB opt-in)
constexpr size_t kPredFixed = 4 * (size_t)kBSpan + kBSpan / 8;      // segment ends + exposed-read flags
constexpr uint32_t kPredCapS = (uint32_t)((kPredSmemS - kPredFixed) / 4);
constexpr uint32_t kPredCapB = (uint32_t)((kPredSmemB - kPredFixed) / 4);

struct PredOut {
  int32_t *pred;                  // [n] last earlier writer of raw iteration i's read (loop-local)
  unsigned long long *V;          // [n] per-iteration shadow slots: V[pred] = 0 for every pred
  uint32_t *pub, *now, *later;    // [nw] each, zeroed by the caller
  int64_t *hdr;                   // H_PRED_FAIL, H_PRED_SEG
  uint32_t *redo;                 // [B] bucket left to the big tier
  const uint32_t *order;          // [B] bucket of CTA k (heaviest first)
  int all_read;                   // SAXPY: every write record also reads its address (Y[w])
};

template <bool BIG>
__device__ __forceinline__ void pred_bucket(int b, const uint32_t *base, const uint32_t *tot,
                                            const unsigned long long *rec, const PredOut &O) {
  constexpr int kT = BIG ? 1024 : 512;
  constexpr uint32_t kCap = BIG ? kPredCapB : kPredCapS;
  extern __shared__ uint32_t s_dyn[];
  // cur[a]: first the writer count of address a, then (scan) the start of its
  // segment, then (fill) its end -- segment a is [cur[a-1], cur[a])
  uint32_t *cur = s_dyn;                    // [kBSpan]
  uint32_t *xflag = cur + kBSpan;           // [kBSpan / 32] address has an exposed read
  uint32_t *wl = xflag + kBSpan / 32;       // [kCap] writer lists
  __shared__ uint32_t s_wsum[kT / 32];
  __shared__ uint32_t s_nw;
  const uint32_t total = tot[b];
  const unsigned long long *rb = rec + base[b];
  for (int k = threadIdx.x; k < kBSpan; k += kT) cur[k] = 0;
  for (int k = threadIdx.x; k < kBSpan / 32; k += kT) xflag[k] = 0;
  __syncthreads();
  constexpr int kU = 4;
  auto sweep = [&](auto &&f) {
    for (uint32_t p0 = threadIdx.x; p0 < total; p0 += kT * kU) {
      unsigned long long xv[kU];
#pragma unroll
      for (int u = 0; u < kU; u++) {
        const uint32_t p = p0 + (uint32_t)u * kT;
        xv[u] = p < total ? rb[p] : 0ull;
      }
#pragma unroll
      for (int u = 0; u < kU; u++)
        if (p0 + (uint32_t)u * kT < total) f(xv[u]);
    }
  };
  sweep([&](unsigned long long x) {
    if (x & kRecW) atomicAdd(&cur[(uint32_t)(x >> 32) & (kBSpan - 1)], 1u);
  });
  __syncthreads();
  // exclusive scan of the counts: kPer addresses per thread
  constexpr int kPer = kBSpan / kT;
  const int a0 = threadIdx.x * kPer;
  uint32_t c[kPer], s = 0, mseg = 0;
#pragma unroll
  for (int k = 0; k < kPer; k++) {
    c[k] = cur[a0 + k];
    s += c[k];
    mseg = max(mseg, c[k]);
  }
  uint32_t x = s;
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
    if ((threadIdx.x & 31) >= o) x += y;
  }
  if ((threadIdx.x & 31) == 31) s_wsum[threadIdx.x >> 5] = x;
  mseg = __reduce_max_sync(0xffffffffu, mseg);
  __syncthreads();
  uint32_t run = x - s;
  for (int k = 0; k < (int)(threadIdx.x >> 5); k++) run += s_wsum[k];
#pragma unroll
  for (int k = 0; k < kPer; k++) {
    cur[a0 + k] = run;
    run += c[k];
  }
  if (threadIdx.x == kT - 1) s_nw = run;
  if ((threadIdx.x & 31) == 0 && mseg)
    atomicMax(reinterpret_cast<unsigned long long *>(&O.hdr[H_PRED_SEG]), (unsigned long long)mseg);
  __syncthreads();
  const uint32_t nwr = s_nw;
  if (nwr == 0) return;   // nothing written in this bucket: no read has a writer
  if (nwr > kCap || __syncthreads_or(mseg > kPredSegCap)) {
    if (threadIdx.x == 0) {
      if (!BIG && nwr > kCap && mseg <= kPredSegCap) O.redo[b] = 1;
      else atomicAdd(reinterpret_cast<unsigned long long *>(&O.hdr[H_PRED_FAIL]), 1ull);
    }
    return;
  }
  sweep([&](unsigned long long x) {
    if (x & kRecW) wl[atomicAdd(&cur[(uint32_t)(x >> 32) & (kBSpan - 1)], 1u)] = (uint32_t)x;
  });
  __syncthreads();
  // reads: the largest writer below i in the address's list
  sweep([&](unsigned long long x) {
    if (!rec_reads(x) && !O.all_read) return;
    const uint32_t i = (uint32_t)x, al = (uint32_t)(x >> 32) & (kBSpan - 1);
    const uint32_t p0 = al ? cur[al - 1] : 0u, p1 = cur[al];
    if (p0 == p1) return;   // an address nobody writes
    uint32_t best = 0xFFFFFFFFu;
    for (uint32_t p = p0; p < p1; p++) {
      const uint32_t j = wl[p];
      if (j < i && (best == 0xFFFFFFFFu || j > best)) best = j;
    }
    if (best != 0xFFFFFFFFu) {
      O.pred[i] = (int32_t)best;
      O.V[best] = 0ull;
      atomicOr(&O.pub[best >> 5], 1u << (best & 31));
    } else {
      atomicOr(&xflag[al >> 5], 1u << (al & 31));
    }
  });
  __syncthreads();
  // writers: the last writer of every written address commits
  for (int al = threadIdx.x; al < kBSpan; al += kT) {
    const uint32_t p0 = al ? cur[al - 1] : 0u, p1 = cur[al];
    if (p0 == p1) continue;
    uint32_t last = wl[p0];
    for (uint32_t p = p0 + 1; p < p1; p++) last = max(last, wl[p]);
    uint32_t *bits = (xflag[al >> 5] >> (al & 31)) & 1u ? O.later : O.now;
    atomicOr(&bits[last >> 5], 1u << (last & 31));
  }
}

__global__ void __launch_bounds__(512, 2) k_bk_pred(const uint32_t *base, const uint32_t *tot,
                                                    const unsigned long long *rec, PredOut O) {
  pred_bucket<false>((int)O.order[blockIdx.x], base, tot, rec, O);
}
// the big tier: one CTA per SM walks the buckets and redoes the marked ones
__global__ void __launch_bounds__(1024, 1) k_bk_pred_big(int B, const uint32_t *base, const uint32_t *tot,
                                                         const unsigned long long *rec, PredOut O) {
  for (int b = blockIdx.x; b < B; b += gridDim.x) {
    if (!O.redo[b]) continue;
    pred_bucket<true>(b, base, tot, rec, O);
    __syncthreads();   // (shared memory reused by the next bucket)
  }
}

// everything the profile accumulates into, reset in one launch: the header
// (first raw iteration = -1), the guide words, the per-chunk counts and the
// per-chunk address ranges (min = ~0, max = 0)
// (with pfx: warp 0 of block 0 also runs the static check's affine sample --
// reading B8: an index array that is not affine on its first m entries is not
// affine -- writes the verdict to hdr[H_GATE] (1: looks affine, the profile's
// kernels queued behind exit at once) and to mapped host words mir[0], then the
// call's sequence number mir[1])
struct PrefixDuty {
  const int32_t *p[4];
  int m;
  long long *mir;
  const volatile unsigned long long *seq;   // the call's sequence number (mapped host word, written before the launch)
};
__global__ void __launch_bounds__(256) k_bk_prep(int64_t *hdr, uint32_t *graw, uint32_t *gsrc, int64_t nw, int64_t *cc,
                                                 int64_t ncc, uint32_t *cr, int64_t nck, PrefixDuty pfx) {
  if (blockIdx.x == 0 && threadIdx.x < 32) {
    bool ok = pfx.m >= 3;
    if (ok)
#pragma unroll
      for (int q = 0; q < 4; q++) {
        if (!pfx.p[q]) continue;
        const int64_t b = __ldg(pfx.p[q]), a = (int64_t)__ldg(pfx.p[q] + 1) - b;
        for (int k = threadIdx.x; k < pfx.m; k += 32) ok = ok && (int64_t)__ldg(pfx.p[q] + k) == b + a * k;
      }
    ok = __all_sync(0xffffffffu, ok);
    if (threadIdx.x == 0) {
      hdr[H_GATE] = ok ? 1 : 0;
      if (pfx.mir) {
        pfx.mir[0] = ok ? 1 : 0;
        asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(pfx.mir + 1), "l"(*pfx.seq) : "memory");
      }
    }
  }
  const int64_t nh = (int64_t)(kHeaderBytes / 8);
  int64_t m = nh;
  if (nw > m) m = nw;
  if (ncc > m) m = ncc;
  if (nck > m) m = nck;
  for (int64_t k = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; k < m; k += (int64_t)gridDim.x * blockDim.x) {
    if (k < nh && k != H_GATE) hdr[k] = k == H_FIRST_RAW ? -1 : 0;
    if (k < nw) {
      if (graw) graw[k] = 0;
      if (gsrc) gsrc[k] = 0;
    }
    if (cc && k < ncc) cc[k] = 0;
    if (cr && k < nck) { cr[2 * k] = 0xFFFFFFFFu; cr[2 * k + 1] = 0u; }
  }
}

namespace {
struct BkPlan {
  BkView v;
  unsigned long long *rec;
  uint32_t *cnt, *tot, *base, *wflag, *order;
};

bool plan(const Job &j, void *ws, const Layout &lo, BkPlan &P) {
  const DLoop &d = j.d;
  if (!ws || d.n <= 0) return false;
  if (j.op == JP_OP_ADD_C) {
    if (!d.r && !d.w) return false;
  } else if (j.op == JP_OP_SAXPY) {
    if (!d.w) return false;
  } else {
    return false;
  }
  if (d.lenA < (1 << 20) || d.lenA > (int64_t)kMaxBuckets * kBSpan) return false;
  if (d.n > (int64_t)kMaxTiles * kTile) return false;
  const char *e = getenv("JP_PROFILE_BUCKETS");
  if (e && e[0] == '0') return false;
  const int B = (int)((d.lenA + kBSpan - 1) / kBSpan), T = (int)((d.n + kTile - 1) / kTile);
  const int64_t nrec = (j.op == JP_OP_ADD_C ? 2 : 1) * d.n;
  // records (8 B each) in minW_A .. keys_A when those regions are contiguous (the
  // profile keeps no tables, and every privatized run clears the keys it
  // applies); offsets in maxRx_A (free until a jp_tls_guide pass, which
  // jp_schedule skips)
  // (the regions follow one another in layout order, separated only by the
  // 256-byte alignment padding of the workspace: the span is one free piece)
  const size_t rb = lo.bytes[R_KEYS_A] ? lo.off[R_KEYS_A] + lo.bytes[R_KEYS_A] - lo.off[R_MINW_A] : 0;
  if (!lo.bytes[R_MINW_A] || rb < 8 * (size_t)nrec) return false;
  if (lo.bytes[R_MAXRX_A] < 4 * ((size_t)T * B + 4 * (size_t)B)) return false;
  // the scatter stages a whole tile plus three words and a flag per bucket in
  // shared memory: len_A up to ~2.7K buckets (~22 M elements) on a 227 KB SM
  static int smax = 0;
  if (!smax) {
    int dev = 0;
    cudaGetDevice(&dev);
    if (cudaDeviceGetAttribute(&smax, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev) != cudaSuccess || smax <= 0) {
      cudaGetLastError();
      smax = 227 * 1024;
    }
  }
  if (6 * 2 * (size_t)kTile + 4 * (3 * (size_t)B + 1) + (size_t)B + 256 > (size_t)smax) return false;
  P.v = BkView{d.r, d.w, d.n, d.ioff, (uint32_t)d.lenA, B, T, nullptr, 1, nullptr};
  P.rec = at<unsigned long long>(ws, lo, R_MINW_A);
  P.cnt = at<uint32_t>(ws, lo, R_MAXRX_A);
  P.tot = P.cnt + (size_t)T * B;
  P.base = P.tot + B;
  P.wflag = P.base + B;
  P.order = P.wflag + B;
  return true;
}

template <int OP>
void run_bucket(const BkPlan &P, const DLoop &d, int64_t *hdr, BkOut O, cudaStream_t st) {
  auto al = [](const int32_t *q) { return q == nullptr || ((uintptr_t)q & 15) == 0; };
  const int vec = al(d.r) && al(d.w);
  const int B = P.v.B, T = P.v.T;
  k_bk_count<OP><<<T, kBThreads, 4 * (size_t)B, st>>>(P.v, vec, P.cnt, &hdr[H_BAD]);
  k_bk_scan_tiles<<<(B + kScanNB - 1) / kScanNB, 1024, 0, st>>>(P.cnt, T, B, P.tot, P.wflag, P.v.gate);
  k_bk_scan_buckets<<<1, 1024, 0, st>>>(P.tot, B, P.base, P.order, P.v.gate);
  const size_t ssm = 6 * 2 * (size_t)kTile + 4 * (3 * (size_t)B + 1) + (size_t)B;
  k_bk_scatter<OP><<<T, kBThreads, ssm, st>>>(P.v, vec, P.cnt, P.tot, P.base, P.wflag, P.rec);
  const int nch = O.cc ? (int)((d.n + O.chunk - 1) / O.chunk) : 0;
  const size_t sm = 4 * (size_t)kBSpan * (OP == JP_OP_ADD_C ? 2 : 1) + (O.cc && nch <= kSmemChunks ? 12 * (size_t)nch : 0);
  k_bk_eval<OP><<<B, kEvalThreads, sm, st>>>(P.v, P.base, P.tot, P.rec, O);
}
// the dynamic shared memory of the scatter and eval kernels, set before any launch
// (and before a stream capture)
template <int OP>
void prepare_bucket(const BkPlan &P, const BkOut &O, const DLoop &d) {
  const int B = P.v.B;
  set_smem_once((const void *)k_bk_scatter<OP>, (int)(6 * 2 * (size_t)kTile + 4 * (3 * (size_t)B + 1) + (size_t)B));
  const int nch = O.cc ? (int)((d.n + O.chunk - 1) / O.chunk) : 0;
  set_smem_once((const void *)k_bk_eval<OP>, (int)(4 * (size_t)kBSpan * (OP == JP_OP_ADD_C ? 2 : 1) +
                                                   (O.cc && nch <= kSmemChunks ? 12 * (size_t)nch : 0)));
}

// The profile's six launches as one CUDA graph per argument set (a call with the
// same loop, workspace and outputs replays it): the host issues one launch instead
// of six (~4-5 us of host time each, which left the GPU idle between the first
// kernels).  Captured on a per-thread side stream, launched into the caller's.
struct BkGraph {
  std::string key;
  cudaGraphExec_t exec;
};
}  // namespace

bool bucket_profile_ok(const Job &j, void *ws, const Layout &lo) {
  BkPlan P;
  return plan(j, ws, lo, P);
}

cudaError_t launch_prof_bucket(const Job &j, void *ws, const Layout &lo, uint32_t *graw, uint32_t *gsrc,
                               int64_t chunk, int64_t *cc, cudaStream_t st, int32_t *wsrc, uint32_t *crange,
                               unsigned long long *vclr, int sample_m, long long *mir,
                               const unsigned long long *seq) {
  BkPlan P;
  if (!plan(j, ws, lo, P)) return cudaErrorInvalidValue;
  PrefixDuty pfx{{j.d.r, j.d.r2, j.d.w, j.d.s}, sample_m, mir, seq};
  if (sample_m > 0 && !seq) return cudaErrorInvalidValue;
  if (sample_m > 0) P.v.gate = &at<int64_t>(ws, lo, R_HEADER)[H_GATE];
  static_assert(kTile == kBucketTile, "jp_host.h kBucketTile");
  int64_t nck = 0;
  if (crange && chunk > 0 && chunk % kTile == 0) {
    nck = (j.d.n + chunk - 1) / chunk;
    P.v.crange = crange;
    P.v.ctiles = (int)(chunk / kTile);
  }
  int64_t *hdr = at<int64_t>(ws, lo, R_HEADER);
  const int64_t nw = (j.d.n + 31) / 32;
  const int64_t ncc = cc ? 3 * ((j.d.n + chunk - 1) / chunk) : 0;
  const int64_t mprep = std::max<int64_t>(std::max<int64_t>((int64_t)(kHeaderBytes / 8), nw), std::max(ncc, nck));
  const int64_t need = (mprep + 255) / 256, cap = (int64_t)num_sms() * 4;
  const int gprep = (int)(need < cap ? need : cap);
  BkOut O{hdr, graw, gsrc, chunk, cc, j.d.base, j.op == JP_OP_ADD_C ? wsrc : nullptr, P.order,
          j.op == JP_OP_ADD_C ? vclr : nullptr};
  if (j.op == JP_OP_ADD_C) prepare_bucket<JP_OP_ADD_C>(P, O, j.d);
  else prepare_bucket<JP_OP_SAXPY>(P, O, j.d);
  auto issue = [&](cudaStream_t s) {
    k_bk_prep<<<gprep, 256, 0, s>>>(hdr, graw, gsrc, nw, cc, ncc, nck ? crange : nullptr, nck, pfx);
    if (j.op == JP_OP_ADD_C) run_bucket<JP_OP_ADD_C>(P, j.d, hdr, O, s);
    else run_bucket<JP_OP_SAXPY>(P, j.d, hdr, O, s);
  };
  note_launch(6);
  const char *ng = getenv("JP_NO_GRAPHS");
  if (ng && ng[0] == '1') {
    issue(st);
    return launch_check();
  }
  int dev = 0;
  cudaGetDevice(&dev);
  // the key: every value the six launches take, field by field (no struct padding)
  std::string key;
  auto put = [&](auto v) { key.append(reinterpret_cast<const char *>(&v), sizeof v); };
  put(dev); put(j.op); put(j.dt); put(gprep); put(nck); put(ncc); put(nw);
  put(P.v.r); put(P.v.w); put(P.v.n); put(P.v.ioff); put(P.v.lenA); put(P.v.B); put(P.v.T); put(P.v.crange);
  put(P.v.ctiles); put(P.v.gate);
  put(P.rec); put(P.cnt); put(P.tot); put(P.base); put(P.wflag); put(P.order);
  put(O.hdr); put(O.graw); put(O.gsrc); put(O.chunk); put(O.cc); put(O.gbase); put(O.wsrc); put(O.order); put(O.vclr);
  for (int q = 0; q < 4; q++) put(pfx.p[q]);
  put(pfx.m); put(pfx.mir); put(pfx.seq);
  put(j.d.r); put(j.d.w); put(j.d.n); put(j.d.ioff); put(j.d.base);
  thread_local std::vector<BkGraph> cache;
  for (const BkGraph &g : cache)
    if (g.key == key) return cudaGraphLaunch(g.exec, st);
  thread_local cudaStream_t cs[64] = {};
  if (!cs[dev & 63]) {
    cudaError_t e = cudaStreamCreateWithFlags(&cs[dev & 63], cudaStreamNonBlocking);
    if (e != cudaSuccess) return e;
  }
  cudaStream_t c = cs[dev & 63];
  cudaError_t e = cudaStreamBeginCapture(c, cudaStreamCaptureModeThreadLocal);
  if (e != cudaSuccess) return e;
  issue(c);
  cudaGraph_t graph = nullptr;
  e = cudaStreamEndCapture(c, &graph);
  if (e != cudaSuccess) return e;
  cudaGraphExec_t exec = nullptr;
  e = cudaGraphInstantiate(&exec, graph, 0);
  cudaGraphDestroy(graph);
  if (e != cudaSuccess) return e;
  if (cache.size() >= 16) {   // (bounded: older argument sets are dropped)
    for (BkGraph &g : cache) cudaGraphExecDestroy(g.exec);
    cache.clear();
  }
  cache.push_back({key, exec});
  return cudaGraphLaunch(exec, st);
}

cudaError_t launch_prof_pred(const Job &j, void *ws, const Layout &lo, int32_t *pred, uint32_t *bits,
                             unsigned long long *V, cudaStream_t st) {
  BkPlan P;
  if ((j.op != JP_OP_ADD_C && j.op != JP_OP_SAXPY) || !plan(j, ws, lo, P)) return cudaErrorInvalidValue;
  const int64_t nw = (j.d.n + 31) / 32;
  cudaError_t e = cudaMemsetAsync(bits, 0, 3 * 4 * (size_t)nw, st);
  // redo flags in the per-tile offsets (P.cnt: the scatter was their last reader)
  if (e == cudaSuccess) e = cudaMemsetAsync(P.cnt, 0, 4 * (size_t)P.v.B, st);
  if (e == cudaSuccess)
    e = set_smem_once((const void *)k_bk_pred, (int)kPredSmemS);
  if (e == cudaSuccess)
    e = set_smem_once((const void *)k_bk_pred_big, (int)kPredSmemB);
  if (e != cudaSuccess) return e;
  PredOut O{pred, V, bits, bits + nw, bits + 2 * nw, at<int64_t>(ws, lo, R_HEADER), P.cnt, P.order,
            j.op == JP_OP_SAXPY};
  k_bk_pred<<<P.v.B, 512, kPredSmemS, st>>>(P.base, P.tot, P.rec, O);
  k_bk_pred_big<<<std::min(P.v.B, num_sms()), 1024, kPredSmemB, st>>>(P.v.B, P.base, P.tot, P.rec, O);
  note_launch(2);
  return launch_check();
}

}  // namespace jp

// jp_priv.cu -- privatized execution PE(V) (the
// private(list) clause, Table I: "a copy of each variable in list is
// allocated for each execution element").
//
// Reading A10: exposed reads see the pre-loop values (legal iff d_raw = 0),
// the covered read of T sees the iteration's own private value (a register).
// Reading A9: after all iterations every address holds the value of its
// highest-gid writer -- realised with packed keys (gid+1)<<32 | bits(v) and
// atomicMax, so it composes across CTAs and (via an int64 MAX all-reduce)
// across GPUs.  Arrays reached only through identity indices are stored
// directly (one writer per address, no key).
//
// Hot-address handling (config 4 writes 2^26 values into 1024 slots): small
// keyed arrays get a per-CTA shared table of the highest local iteration that
// wrote each slot.  Each CTA walks its iterations in DESCENDING order, so the
// first touch of a slot is already its CTA-local last writer and every later
// touch fails the plain shared-memory check without issuing an atomic; the
// flush then recomputes the winner's value and issues one 64-bit global
// atomicMax per (CTA, touched slot).
#include <cooperative_groups.h>
#include <atomic>
#include <cstring>
#include "jp_host.h"

namespace cg = cooperative_groups;

namespace jp {

constexpr int kPrivThreads = 512;

__device__ __forceinline__ void smem_last(uint32_t *tab, int64_t a, int64_t i) {
  const uint32_t v = (uint32_t)(i + 1);
  if (tab[a] < v) atomicMax(&tab[a], v);
}

template <int OP, int DT>
__global__ void __launch_bounds__(kPrivThreads) k_priv_generic(DLoop L, unsigned long long *kA,
                                                                unsigned long long *kT, int smA, int smT) {
  if (aborted(L)) return;
  extern __shared__ uint32_t sm[];
  uint32_t *tA = smA ? sm : nullptr;
  uint32_t *tT = smT ? sm + (smA ? L.lenA : 0) : nullptr;
  const int64_t ns = (smA ? L.lenA : 0) + (smT ? L.lenT : 0);
  for (int64_t k = threadIdx.x; k < ns; k += blockDim.x) sm[k] = 0;
  JP_CTA_SYNC();
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t j = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; j < L.n; j += stride) {
    const int64_t i = L.n - 1 - j;          // descending within every CTA
    uint32_t va = 0, vt = 0;
    body_values<OP, DT>(L, i, L.A, va, vt);  // A is untouched until finalize when keyed
    const int64_t a = ixl(L, L.w, i);
    if (kA) {
      if (tA) smem_last(tA, a, i);
      else atomicMax(&kA[a], pack_key(L.base + i, va));
    } else {
      L.A[a] = va;
    }
    if constexpr (OP == JP_OP_PRIV_TMP) {
      const int64_t b = ixl(L, L.s, i);
      if (kT) {
        if (tT) smem_last(tT, b, i);
        else atomicMax(&kT[b], pack_key(L.base + i, vt));
      } else {
        L.T[b] = vt;
      }
    }
  }
  JP_CTA_SYNC();
  if (tA) {
    for (int64_t a = threadIdx.x; a < L.lenA; a += blockDim.x) {
      const uint32_t e = tA[a];
      if (e) {
        uint32_t va = 0, vt = 0;
        body_values<OP, DT>(L, e - 1, L.A, va, vt);
        atomicMax(&kA[a], pack_key(L.base + e - 1, va));
      }
    }
  }
  if (tT) {
    for (int64_t b = threadIdx.x; b < L.lenT; b += blockDim.x) {
      const uint32_t e = tT[b];
      if (e) {
        uint32_t va = 0, vt = 0;
        body_values<OP, DT>(L, e - 1, L.A, va, vt);
        atomicMax(&kT[b], pack_key(L.base + e - 1, vt));
      }
    }
  }
}

// PRIV_TMP with r = w = NULL, s indirect, small T (config 4): 16-byte lanes.
// Per iteration: X 4 B + s 4 B read, Y 4 B written (12 B/iter algorithmic).
template <int DT>
__global__ void __launch_bounds__(kPrivThreads) k_priv_tmp_vec(DLoop L, unsigned long long *kT, int64_t nvec) {
  if (aborted(L)) return;
  extern __shared__ uint32_t tT[];
  for (int64_t k = threadIdx.x; k < L.lenT; k += blockDim.x) tT[k] = 0;
  JP_CTA_SYNC();
  const uint4 *X4 = reinterpret_cast<const uint4 *>(L.X);
  const int4 *S4 = reinterpret_cast<const int4 *>(L.s);
  uint4 *Y4 = reinterpret_cast<uint4 *>(L.A);
  constexpr int U = 2;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x * U;
  for (int64_t j0 = (int64_t)blockIdx.x * blockDim.x * U + threadIdx.x; j0 < nvec; j0 += stride) {
    uint4 x[U];
    int4 s[U];
#pragma unroll
    for (int u = 0; u < U; u++) {
      const int64_t j = j0 + (int64_t)u * blockDim.x;
      if (j < nvec) {
        const int64_t v = nvec - 1 - j;
        x[u] = __ldcs(X4 + v);
        s[u] = __ldcs(S4 + v);
      }
    }
#pragma unroll
    for (int u = 0; u < U; u++) {
      const int64_t j = j0 + (int64_t)u * blockDim.x;
      if (j < nvec) {
        const int64_t v = nvec - 1 - j;
        uint4 y;
        y.x = op_add<DT>(op_mul<DT>(L.c0, x[u].x), L.c1);
        y.y = op_add<DT>(op_mul<DT>(L.c0, x[u].y), L.c1);
        y.z = op_add<DT>(op_mul<DT>(L.c0, x[u].z), L.c1);
        y.w = op_add<DT>(op_mul<DT>(L.c0, x[u].w), L.c1);
        __stcs(Y4 + v, y);
        smem_last(tT, s[u].w, 4 * v + 3);
        smem_last(tT, s[u].z, 4 * v + 2);
        smem_last(tT, s[u].y, 4 * v + 1);
        smem_last(tT, s[u].x, 4 * v + 0);
      }
    }
  }
  if (blockIdx.x == 0) {  // scalar tail [4*nvec, n)
    for (int64_t i = 4 * nvec + threadIdx.x; i < L.n; i += blockDim.x) {
      const uint32_t t = op_mul<DT>(L.c0, L.X[i]);
      L.A[i] = op_add<DT>(t, L.c1);
      smem_last(tT, L.s[i], i);
    }
  }
  JP_CTA_SYNC();
  for (int64_t b = threadIdx.x; b < L.lenT; b += blockDim.x) {
    const uint32_t e = tT[b];
    if (e) atomicMax(&kT[b], pack_key(L.base + e - 1, op_mul<DT>(L.c0, L.X[e - 1])));
  }
}

// Same loop, bulk-copy (TMA) staged: one CTA per SM walks its tiles in
// DESCENDING order through a kPrivStages ring of {X, s} 16 KiB tiles (mbarrier
// completion), computes Y in place of X in shared memory and bulk-stores it;
// the slot table is updated from the staged s tile (descending inside the tile
// too, so the check-before-atomic filter keeps working).
constexpr int kPrivTile = 4096, kPrivStages = 4, kPrivTmaThreads = 256;

// (k_priv_tmp_tma is the one-pass stream whose keys are merged by a later C4 and
// finalize; R1 + R2 in one launch is k_priv_tmp_2ph below.)
// C4 fused into the stream (jp_priv_stream_merge): every rank's inbox holds
//   [0] epoch of the last merge, [32 + 2*8] flags[parity][sender] = epoch,
//   [64 ...] keys[parity][sender][lenT]
// and every rank maps every rank's inbox (CUDA IPC / NVLink peer memory).
constexpr int kMergePeers = 8;
constexpr int64_t kInboxFlags = 32, kInboxKeys = 64;
struct MergeP2P {
  unsigned long long *inbox[kMergePeers];   // every rank's inbox, mapped here (own included)
  int world, me;
  int *err;
};

__device__ __forceinline__ unsigned long long gtimer_ns() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}

// One CTA, after the grid barrier that follows every CTA's key flush: push this
// rank's keys into slot (parity, me) of every rank's inbox with plain peer
// stores (posted over NVLink), a system fence, then one release flag per peer;
// wait for every sender's flag of this epoch in the local inbox; reduce the
// world key tables (local loads) and apply the merged last writers to T.
// Double-buffered by epoch parity: a rank writes parity e+1 only after its
// merge e, which needed every peer's flag e, i.e. every peer's push e -- pushes
// of e+1 never land in a buffer a peer still reduces for e-1.
struct MergeState { unsigned long long e; int par; };

// push this rank's keys into slot (parity, me) of every rank's inbox and raise
// one system-scope release flag per peer (CTA 0, all keys in kT)
__device__ MergeState merge_p2p_push(const DLoop &L, const unsigned long long *kT, const MergeP2P &M) {
  __shared__ unsigned long long e_s;
  unsigned long long *in = M.inbox[M.me];
  const int tid = threadIdx.x, nt = blockDim.x;
  const int64_t lenT = L.lenT;
  if (tid == 0) e_s = in[0] + 1;
  __syncthreads();
  const unsigned long long e = e_s;
  const int par = (int)(e & 1);
  for (int p = 0; p < M.world; p++) {
    unsigned long long *dst = M.inbox[p] + kInboxKeys + ((int64_t)par * M.world + M.me) * lenT;
    for (int64_t b = tid; b < lenT; b += nt) dst[b] = __ldcg(kT + b);
  }
  // the CTA barrier orders every thread's pushes before the flag writers'
  // system-scope release (cumulative): no fence per pushing thread
  __syncthreads();
  if (tid < M.world) {
    unsigned long long *f = M.inbox[tid] + kInboxFlags + par * kMergePeers + M.me;
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(f), "l"(e) : "memory");
  }
  return MergeState{e, par};
}

// wait for every sender's flag of this epoch, reduce the world tables (local
// loads) and apply the merged last writers to T (CTA 0)
__device__ void merge_p2p_finish(const DLoop &L, const MergeP2P &M, MergeState st) {
  __shared__ int ok;
  unsigned long long *in = M.inbox[M.me];
  const int tid = threadIdx.x, nt = blockDim.x;
  const int64_t lenT = L.lenT;
  if (tid == 0) ok = 1;
  __syncthreads();
  if (tid < M.world) {
    const unsigned long long *g = in + kInboxFlags + st.par * kMergePeers + tid;
    const unsigned long long t0 = gtimer_ns();
    for (;;) {
      unsigned long long v;
      asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(g) : "memory");
      if (v >= st.e) break;
      if (gtimer_ns() - t0 > 4000000000ull) { ok = 0; atomicExch(M.err, 1); break; }
      __nanosleep(100);
    }
  }
  __syncthreads();
  if (!ok) return;
  asm volatile("fence.acq_rel.sys;" ::: "memory");
  const unsigned long long *keys = in + kInboxKeys + (int64_t)st.par * M.world * lenT;
  for (int64_t b = tid; b < lenT; b += nt) {
    unsigned long long m = 0;
    for (int r = 0; r < M.world; r++) {
      const unsigned long long v = __ldcv(keys + (int64_t)r * lenT + b);
      m = v > m ? v : m;
    }
    if (m) L.T[b] = (uint32_t)m;
  }
  __syncthreads();
  if (tid == 0) in[0] = st.e;
}

// One CTA, after the grid barrier that follows every CTA's key flush: push this
// rank's keys into slot (parity, me) of every rank's inbox with plain peer
// stores (posted over NVLink), then one release flag per peer; wait for every
// sender's flag of this epoch in the local inbox; reduce the world key tables
// (local loads) and apply the merged last writers to T.  Double-buffered by
// epoch parity: a rank writes parity e+1 only after its merge e, which needed
// every peer's flag e, i.e. every peer's push e -- pushes of e+1 never land in
// a buffer a peer still reduces for e-1.
__device__ void merge_p2p_epilogue(const DLoop &L, const unsigned long long *kT, const MergeP2P &M) {
  merge_p2p_finish(L, M, merge_p2p_push(L, kT, M));
}

// Two phases in one cooperative kernel (config-4 shape, the whole call's run):
// phase 1 streams s alone -- the index check of reading A13 (out-of-range slots
// counted into *vbad, nullable) and the per-CTA last-writer table, flushed as
// packed keys (the value c0*X[i] recomputed at the CTA's last writer of a slot);
// a grid barrier; then, only if no index was bad, phase 2 streams X into Y =
// c0*X + c1 and every CTA applies a slice of the keys to T.  s, X and Y each
// cross HBM once: 12 B/iter, the check included.
// 4 stages of 32 KiB per phase (the same 128 KiB of shared memory as the one-pass
// kernel): 16 KiB tiles left each CTA bound by its per-tile barrier / bulk-store
// turnaround in the X -> Y phase (188 us for config 4, ncu)
constexpr int kPh = kPrivStages, kPh2Tile = 2 * kPrivTile, kPh2Threads = 1024;
template <int DT>
__global__ void __launch_bounds__(kPh2Threads, 1) k_priv_tmp_2ph(DLoop L, unsigned long long *kT, int64_t ntiles,
                                                                     int64_t *vbad, int64_t *mirror,
                                                                     unsigned long long seq) {
  extern __shared__ __align__(128) uint32_t psm[];   // [kPh][tile] then tT[lenT]
  __shared__ __align__(8) unsigned long long full1[kPh], full2[kPh];
  uint32_t *tT = psm + (size_t)kPh * kPh2Tile;
  const int tid = threadIdx.x;
  const uint32_t lenT = (uint32_t)L.lenT;
  for (int64_t k = tid; k < L.lenT; k += kPh2Threads) tT[k] = 0;
  // the key table and the index-error count are cleared here (no memset
  // launches ahead of the kernel); the grid barrier after phase 1 orders the
  // clears before every CTA's flush
  for (int64_t b = (int64_t)blockIdx.x * kPh2Threads + tid; b < L.lenT; b += (int64_t)gridDim.x * kPh2Threads)
    kT[b] = 0;
  if (vbad && blockIdx.x == 0 && tid == 0) *vbad = 0;
  const int64_t my = ntiles > blockIdx.x ? (ntiles - 1 - blockIdx.x) / gridDim.x + 1 : 0;
  auto tile_of = [&](int64_t k) { return ntiles - 1 - (int64_t)blockIdx.x - k * gridDim.x; };
  auto buf = [&](int64_t k) { return psm + (size_t)(k % kPh) * kPh2Tile; };
  if (tid == 0) {
    for (int sg = 0; sg < kPh; sg++) { mbar_init(&full1[sg], 1); mbar_init(&full2[sg], 1); }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  // ---------------- phase 1: s ----------------
  auto issue1 = [&](int64_t k) {
    mbar_expect_tx(&full1[k % kPh], kPh2Tile * 4);
    bulk_load(buf(k), L.s + tile_of(k) * kPh2Tile, kPh2Tile * 4, &full1[k % kPh]);
  };
  if (tid == 0)
    for (int64_t k = 0; k < kPh && k < my; k++) issue1(k);
  unsigned bad = 0;
  bool full = false;   // this CTA's slot table has a writer in every slot
  for (int64_t k = 0; k < my; k++) {
    mbar_wait(&full1[k % kPh], (uint32_t)((k / kPh) & 1));
    const int64_t e0 = tile_of(k) * kPh2Tile;
    const int4 *S4 = reinterpret_cast<const int4 *>(buf(k));
    // the slot table's current values are read for all of a thread's iterations
    // first, then the (rare, with the descending walk) atomics issued: a stale
    // read only costs an extra atomicMax, and the loads no longer wait behind
    // possibly aliasing atomics one by one
    constexpr int kQ = kPh2Tile / 4 / kPh2Threads;
    int sl[4 * kQ];
    uint32_t cur[4 * kQ];
#pragma unroll
    for (int q = 0; q < kQ; q++) {
      const int4 sv = S4[kPh2Tile / 4 - 1 - (q * kPh2Threads + tid)];   // descending in the tile
      sl[4 * q + 0] = sv.w; sl[4 * q + 1] = sv.z; sl[4 * q + 2] = sv.y; sl[4 * q + 3] = sv.x;
    }
    if (full) {
      // every slot already has a writer from a later tile of this CTA (tiles are
      // walked in descending order): this tile only needs the index check
#pragma unroll
      for (int m = 0; m < 4 * kQ; m++) bad += (uint32_t)sl[m] >= lenT;
    } else {
#pragma unroll
      for (int m = 0; m < 4 * kQ; m++) {
        const bool ok = (uint32_t)sl[m] < lenT;
        bad += !ok;
        cur[m] = ok ? tT[sl[m]] : 0xFFFFFFFFu;
      }
#pragma unroll
      for (int m = 0; m < 4 * kQ; m++) {
        const int q = m >> 2;
        const int64_t i = e0 + 4 * (kPh2Tile / 4 - 1 - (q * kPh2Threads + tid)) + (3 - (m & 3));
        const uint32_t v = (uint32_t)(i + 1);
        if (cur[m] < v) atomicMax(&tT[sl[m]], v);
      }
      __syncthreads();
      // a slot table this CTA has filled stays filled: later (lower) tiles of the
      // CTA cannot hold a last writer (the coupon collector: 1024 slots are all
      // seen within a tile or two of config 4's random s)
      bool mine = true;
      for (int64_t b = tid; b < (int64_t)lenT; b += kPh2Threads) mine = mine && tT[b] != 0;
      full = __syncthreads_count(mine) == kPh2Threads;
    }
    __syncthreads();   // the stage is read: refill it
    if (tid == 0 && k + kPh < my) issue1(k + kPh);
  }
  if (blockIdx.x == 0)   // element tail [ntiles * tile, n)
    for (int64_t i = ntiles * kPh2Tile + tid; i < L.n; i += kPh2Threads) {
      const int32_t sv = L.s[i];
      if ((uint32_t)sv < lenT) smem_last(tT, sv, i); else bad++;
    }
  bad = __reduce_add_sync(0xffffffffu, bad);
  cg::this_grid().sync();   // the clears above are visible to every CTA
  if (vbad && (tid & 31) == 0 && bad) atomicAdd(reinterpret_cast<unsigned long long *>(vbad), (unsigned long long)bad);
  for (int64_t b = tid; b < L.lenT; b += kPh2Threads) {
    const uint32_t e = tT[b];
    if (e) atomicMax(&kT[b], pack_key(L.base + e - 1, op_mul<DT>(L.c0, __ldg(L.X + e - 1))));
  }
  cg::this_grid().sync();   // every CTA's keys are in, every index checked
  const int64_t nbad = vbad ? *reinterpret_cast<volatile int64_t *>(vbad) : 0;
  if (mirror && blockIdx.x == 0 && tid == 0) {
    // the count to mapped host memory, then the call's sequence number: the
    // host returns as soon as it sees it (the X -> Y phase is stream-ordered)
    mirror[0] = nbad;
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(mirror + 1), "l"(seq) : "memory");
  }
  if (nbad) return;   // nothing written (reading A13)
  for (int64_t b = (int64_t)blockIdx.x * kPh2Threads + tid; b < L.lenT; b += (int64_t)gridDim.x * kPh2Threads) {
    const unsigned long long key = __ldcg(&kT[b]);
    if (key) L.T[b] = (uint32_t)key;
  }
  // ---------------- phase 2: X -> Y ----------------
  auto issue2 = [&](int64_t k) {
    mbar_expect_tx(&full2[k % kPh], kPh2Tile * 4);
    bulk_load(buf(k), L.X + tile_of(k) * kPh2Tile, kPh2Tile * 4, &full2[k % kPh]);
  };
  if (tid == 0)
    for (int64_t k = 0; k < kPh - 1 && k < my; k++) issue2(k);
  for (int64_t k = 0; k < my; k++) {
    mbar_wait(&full2[k % kPh], (uint32_t)((k / kPh) & 1));
    uint4 *X4 = reinterpret_cast<uint4 *>(buf(k));
#pragma unroll
    for (int q = 0; q < kPh2Tile / 4 / kPh2Threads; q++) {
      const int v = q * kPh2Threads + tid;
      const uint4 x = X4[v];
      uint4 y;
      y.x = op_add<DT>(op_mul<DT>(L.c0, x.x), L.c1);
      y.y = op_add<DT>(op_mul<DT>(L.c0, x.y), L.c1);
      y.z = op_add<DT>(op_mul<DT>(L.c0, x.z), L.c1);
      y.w = op_add<DT>(op_mul<DT>(L.c0, x.w), L.c1);
      X4[v] = y;
    }
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    __syncthreads();
    if (tid == 0) {
      bulk_store(L.A + tile_of(k) * kPh2Tile, buf(k), kPh2Tile * 4);
      asm volatile("cp.async.bulk.commit_group;" ::: "memory");
      if (k + kPh - 1 < my) {
        asm volatile("cp.async.bulk.wait_group.read 1;" ::: "memory");
        issue2(k + kPh - 1);
      }
    }
  }
  if (tid == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
  if (blockIdx.x == 0)
    for (int64_t i = ntiles * kPh2Tile + tid; i < L.n; i += kPh2Threads)
      L.A[i] = op_add<DT>(op_mul<DT>(L.c0, L.X[i]), L.c1);
}

// fuse_apply (cooperative launch): after every CTA's flush a grid barrier, then
// the keys are applied to T by every CTA (R1 + R2 in one launch when the index
// check is not needed; k_priv_tmp_2ph carries the check)
template <int DT, bool MERGE = false>
__global__ void __launch_bounds__(kPrivTmaThreads, 1) k_priv_tmp_tma(DLoop L, unsigned long long *kT, int64_t ntiles,
                                                                     int fuse_apply, MergeP2P M = MergeP2P{}) {
  if (aborted(L)) return;
  extern __shared__ __align__(128) uint32_t psm[];   // [stage][2][tile] then tT[lenT]
  __shared__ __align__(8) unsigned long long full[kPrivStages];
  uint32_t *tT = psm + (size_t)kPrivStages * 2 * kPrivTile;
  const int tid = threadIdx.x;
  for (int64_t k = tid; k < L.lenT; k += kPrivTmaThreads) tT[k] = 0;
  // this CTA's tiles, highest first: t = ntiles-1-blockIdx.x - k*gridDim.x
  const int64_t my = ntiles > blockIdx.x ? (ntiles - 1 - blockIdx.x) / gridDim.x + 1 : 0;
  auto tile_of = [&](int64_t k) { return ntiles - 1 - (int64_t)blockIdx.x - k * gridDim.x; };
  auto issue = [&](int64_t k) {
    const int sg = (int)(k % kPrivStages);
    const int64_t e0 = tile_of(k) * kPrivTile;
    uint32_t *bX = psm + (size_t)sg * 2 * kPrivTile, *bS = bX + kPrivTile;
    mbar_expect_tx(&full[sg], 2 * kPrivTile * 4);
    bulk_load(bX, L.X + e0, kPrivTile * 4, &full[sg]);
    bulk_load(bS, L.s + e0, kPrivTile * 4, &full[sg]);
  };
  if (tid == 0) {
    for (int sg = 0; sg < kPrivStages; sg++) mbar_init(&full[sg], 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  if (tid == 0)
    for (int64_t k = 0; k < kPrivStages - 1 && k < my; k++) issue(k);
  for (int64_t k = 0; k < my; k++) {
    const int sg = (int)(k % kPrivStages);
    uint32_t *bX = psm + (size_t)sg * 2 * kPrivTile, *bS = bX + kPrivTile;
    mbar_wait(&full[sg], (uint32_t)((k / kPrivStages) & 1));
    const int64_t e0 = tile_of(k) * kPrivTile;
    uint4 *X4 = reinterpret_cast<uint4 *>(bX);
    const int4 *S4 = reinterpret_cast<const int4 *>(bS);
#pragma unroll
    for (int q = 0; q < kPrivTile / 4 / kPrivTmaThreads; q++) {
      const int v = kPrivTile / 4 - 1 - (q * kPrivTmaThreads + tid);   // descending in the tile
      const uint4 x = X4[v];
      const int4 sv = S4[v];
      uint4 y;
      y.x = op_add<DT>(op_mul<DT>(L.c0, x.x), L.c1);
      y.y = op_add<DT>(op_mul<DT>(L.c0, x.y), L.c1);
      y.z = op_add<DT>(op_mul<DT>(L.c0, x.z), L.c1);
      y.w = op_add<DT>(op_mul<DT>(L.c0, x.w), L.c1);
      X4[v] = y;
      const int64_t i0 = e0 + 4 * v;
      smem_last(tT, sv.w, i0 + 3);
      smem_last(tT, sv.z, i0 + 2);
      smem_last(tT, sv.y, i0 + 1);
      smem_last(tT, sv.x, i0 + 0);
    }
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    __syncthreads();
    if (tid == 0) {
      bulk_store(L.A + e0, bX, kPrivTile * 4);
      asm volatile("cp.async.bulk.commit_group;" ::: "memory");
      if (k + kPrivStages - 1 < my) {
        asm volatile("cp.async.bulk.wait_group.read 1;" ::: "memory");
        issue(k + kPrivStages - 1);
      }
    }
  }
  if (tid == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
  if (blockIdx.x == 0) {   // element tail [ntiles * tile, n)
    for (int64_t i = ntiles * kPrivTile + tid; i < L.n; i += kPrivTmaThreads) {
      L.A[i] = op_add<DT>(op_mul<DT>(L.c0, L.X[i]), L.c1);
      smem_last(tT, L.s[i], i);
    }
  }
  __syncthreads();
  for (int64_t b = tid; b < L.lenT; b += kPrivTmaThreads) {
    const uint32_t e = tT[b];
    if (e) atomicMax(&kT[b], pack_key(L.base + e - 1, op_mul<DT>(L.c0, L.X[e - 1])));
  }
  if (fuse_apply) {
    cg::this_grid().sync();   // every CTA's keys are in
    if constexpr (MERGE) {   // C4 across the ranks and R2, by CTA 0 (jp_priv_stream_merge)
      if (blockIdx.x == 0) merge_p2p_epilogue(L, kT, M);
      return;
    }
    for (int64_t b = (int64_t)blockIdx.x * kPrivTmaThreads + tid; b < L.lenT; b += (int64_t)gridDim.x * kPrivTmaThreads) {
      const unsigned long long k = __ldcg(&kT[b]);
      if (k) L.T[b] = (uint32_t)k;
    }
  }
}

__global__ void k_apply_keys(uint32_t *arr, int64_t len, const unsigned long long *keys, const int64_t *abort) {
  if (abort && *reinterpret_cast<const volatile int64_t *>(abort)) return;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t a = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; a < len; a += stride) {
    const unsigned long long k = keys[a];
    if (k) arr[a] = (uint32_t)k;   // written only where some iteration wrote (safe beside concurrent tasks)
  }
}

static bool al16(const void *p) { return ((uintptr_t)p & 15) == 0; }

template <int OP, int DT>
static void run_priv(const DLoop &d0, unsigned long long *kA, unsigned long long *kT, cudaStream_t st, int max_ctas,
                     bool fuse_apply, bool *applied, int64_t *vbad, bool clear_keys, int64_t *mirror,
                     unsigned long long seq, bool *published) {
  // the key tables start at zero: cleared here, except by the two-phase kernel
  // (which clears its table itself)
  auto clear = [&]() {
    if (!clear_keys) return;
    if (kA) cudaMemsetAsync(kA, 0, 8 * (size_t)d0.lenA, st);
    if (kT) cudaMemsetAsync(kT, 0, 8 * (size_t)d0.lenT, st);
  };
  // vbad: validate the indirect indices first (reading A13), one streaming pass
  // ahead of the run (an in-kernel phase before a grid barrier was measured
  // slower: 177 vs ~169 us device time on config 4); the stream kernels then
  // exit at once on a nonzero count (d0.abort == vbad)
  auto validate_first = [&]() {
    if (vbad) launch_validate_indirect(Job{d0, OP, DT}, vbad, st);
  };
  int grid = num_sms() * 2;
  if (max_ctas > 0 && grid > max_ctas) grid = max_ctas;
  if constexpr (OP == JP_OP_PRIV_TMP) {
    // a rank-local range (B1): X and Y are reached only through identity
    // indices, so rebase them to the range's first element
    DLoop d = d0;
    if (!d.r && !d.w && d.ioff > 0) {
      d.X += d.ioff; d.lenX -= d.ioff;
      d.A += d.ioff; d.lenA -= d.ioff;
      d.ioff = 0;
    }
    if (!d.r && !d.w && d.s && d.ioff == 0 && kT && !kA && d.lenT <= kSmemSlots && al16(d.X) && al16(d.s) &&
        al16(d.A)) {
      if (doall_kernel_choice() == 1) {   // bulk-copy staged (the DOALL kernel choice covers both streams)
        const int64_t ntiles = d.n / kPrivTile;
        const size_t smem = (size_t)kPrivStages * 2 * kPrivTile * 4 + (size_t)d.lenT * 4;
        set_smem_once((const void *)k_priv_tmp_tma<DT>, (int)smem);
        int g = num_sms();
        if (max_ctas > 0 && g > max_ctas) g = max_ctas;
        if (ntiles < g) g = (int)(ntiles < 1 ? 1 : ntiles);
        if (fuse_apply && !vbad) {   // R1 + R2 in one pass (cooperative: one CTA per SM, co-resident)
          clear();
          DLoop dd = d;
          int64_t nt = ntiles;
          int fuse = 1;
          MergeP2P none{};
          void *args[] = {&dd, &kT, &nt, &fuse, &none};
          cudaLaunchCooperativeKernel((void *)k_priv_tmp_tma<DT>, dim3(g), dim3(kPrivTmaThreads), args, smem, st);
          *applied = true;
        } else if (fuse_apply) {   // with the index check: two phases (s, then X -> Y)
          const int64_t ntiles = d.n / kPh2Tile;
          int g = num_sms();
          if (max_ctas > 0 && g > max_ctas) g = max_ctas;
          if (ntiles < g) g = (int)(ntiles < 1 ? 1 : ntiles);
          // two phases: s (index check + last writers), grid barrier, X -> Y and T;
          // the check of reading A13 needs no pass of its own (s crosses HBM once)
          DLoop dd = d;
          dd.abort = nullptr;
          int64_t nt = ntiles;
          int64_t *vb = vbad;
          int64_t *mir = mirror;
          unsigned long long sq = seq;
          void *args[] = {&dd, &kT, &nt, &vb, &mir, &sq};
          // one dynamic-smem limit for every call (lenT <= kSmemSlots), set once per device
          static std::atomic<unsigned long long> attr{0};
          int dev = 0;
          cudaGetDevice(&dev);
          const unsigned long long bit = 1ull << (dev & 63);
          if (!(attr.load() & bit)) {
            const size_t smax = (size_t)kPh * kPh2Tile * 4 + (size_t)kSmemSlots * 4;
            if (set_smem_once((const void *)k_priv_tmp_2ph<DT>, (int)smax) ==
                cudaSuccess)
              attr.fetch_or(bit);
          }
          cudaLaunchCooperativeKernel((void *)k_priv_tmp_2ph<DT>, dim3(g), dim3(kPh2Threads), args, smem, st);
          *applied = true;
          if (published) *published = mirror != nullptr;
        } else {
          clear();
          validate_first();
          k_priv_tmp_tma<DT><<<g, kPrivTmaThreads, smem, st>>>(d, kT, ntiles, 0, MergeP2P{});
        }
        note_launch();
        return;
      }
      int64_t nvec = d.n / 4;
      int64_t need = (nvec + kPrivThreads * 2 - 1) / (kPrivThreads * 2);
      if (need < grid) grid = (int)(need < 1 ? 1 : need);
      clear();
      validate_first();
      k_priv_tmp_vec<DT><<<grid, kPrivThreads, d.lenT * 4, st>>>(d, kT, nvec);
      note_launch();
      return;
    }
  }
  const DLoop &d = d0;
  int smA = kA && d.lenA <= kSmemSlots, smT = kT && d.lenT <= kSmemSlots;
  size_t smem = ((smA ? d.lenA : 0) + (smT ? d.lenT : 0)) * 4;
  int64_t need = (d.n + kPrivThreads - 1) / kPrivThreads;
  if (need < grid) grid = (int)(need < 1 ? 1 : need);
  clear();
  validate_first();
  k_priv_generic<OP, DT><<<grid, kPrivThreads, smem, st>>>(d, kA, kT, smA, smT);
  note_launch();
}

bool priv_merge_ok(const Job &j, int world) {
  const DLoop &d = j.d;
  return j.op == JP_OP_PRIV_TMP && !d.r && !d.w && d.s && d.lenT > 0 && d.lenT <= kSmemSlots && world >= 1 &&
         world <= kMergePeers && al16(d.X + d.ioff) && al16(d.s) && al16(d.A + d.ioff);
}

size_t priv_inbox_bytes(const Job &j, int world) {
  return priv_merge_ok(j, world) ? 8 * ((size_t)kInboxKeys + 2 * (size_t)world * (size_t)j.d.lenT) : 0;
}

cudaError_t launch_priv_stream_merge(const Job &j, unsigned long long *kT, unsigned long long *const *inbox, int world,
                                     int me, int *err, cudaStream_t st) {
  DLoop d = j.d;   // rank-local range (B1): X and Y rebased to the range's first element
  d.X += d.ioff; d.lenX -= d.ioff;
  d.A += d.ioff; d.lenA -= d.ioff;
  d.ioff = 0;
  cudaMemsetAsync(kT, 0, 8 * (size_t)d.lenT, st);
  // the one-pass stream (the ranks' indices were checked by the partitioned
  // profile) with the merge as its epilogue: measured faster than merging from
  // the two-phase kernel, whose s-only phase costs more than the overlap of the
  // exchange with the Y stream saves
  const int64_t ntiles = d.n / kPrivTile;
  const size_t smem = (size_t)kPrivStages * 2 * kPrivTile * 4 + (size_t)d.lenT * 4;
  cudaError_t e;
  auto go = [&](auto kern) {
    set_smem_once((const void *)kern, (int)smem);
    int g = num_sms();
    if (ntiles < g) g = (int)(ntiles < 1 ? 1 : ntiles);
    MergeP2P M{};
    for (int k = 0; k < world; k++) M.inbox[k] = inbox[k];
    M.world = world;
    M.me = me;
    M.err = err;
    int64_t nt = ntiles;
    int fuse = 1;
    void *args[] = {&d, &kT, &nt, &fuse, &M};
    e = cudaLaunchCooperativeKernel((const void *)kern, dim3(g), dim3(kPrivTmaThreads), args, smem, st);
  };
  if (j.dt == JP_F32) go(k_priv_tmp_tma<JP_F32, true>);
  else go(k_priv_tmp_tma<JP_I32, true>);
  note_launch();
  if (e != cudaSuccess) return e;
  return launch_check();
}

cudaError_t launch_priv_stream(const Job &j, void *ws, const Layout &lo, bool clear_keys, cudaStream_t st,
                               int max_ctas, bool fuse_apply, bool *applied, int64_t *validate, int64_t *mirror,
                               unsigned long long seq, bool *published) {
  bool dummy = false, dummy2 = false;
  if (!applied) applied = &dummy;
  if (!published) published = &dummy2;
  *applied = false;
  *published = false;
  auto *kA = at<unsigned long long>(ws, lo, R_KEYS_A);
  auto *kT = at<unsigned long long>(ws, lo, R_KEYS_T);
  if (j.d.n == 0) {
    if (clear_keys) {
      if (kA) cudaMemsetAsync(kA, 0, lo.bytes[R_KEYS_A], st);
      if (kT) cudaMemsetAsync(kT, 0, lo.bytes[R_KEYS_T], st);
    }
    if (validate) cudaMemsetAsync(validate, 0, sizeof(int64_t), st);
    return launch_check();
  }
  JP_DISPATCH(j.op, j.dt, run_priv, j.d, kA, kT, st, max_ctas, fuse_apply, applied, validate, clear_keys, mirror, seq,
              published);
  return launch_check();
}

static void apply(uint32_t *arr, int64_t len, const unsigned long long *keys, cudaStream_t st,
                  const int64_t *abort = nullptr) {
  if (!len || !keys) return;
  int64_t need = (len + 255) / 256, cap = (int64_t)num_sms() * 8;
  k_apply_keys<<<(int)(need < cap ? need : cap), 256, 0, st>>>(arr, len, keys, abort);
  note_launch();
}

cudaError_t launch_priv_finalize(const Job &j, void *ws, const Layout &lo, cudaStream_t st) {
  apply(j.d.A, j.d.lenA, at<unsigned long long>(ws, lo, R_KEYS_A), st, j.d.abort);
  if (j.op == JP_OP_PRIV_TMP) apply(j.d.T, j.d.lenT, at<unsigned long long>(ws, lo, R_KEYS_T), st, j.d.abort);
  return launch_check();
}

// Packed last-writer keys of what a loop (or a range of one) has ALREADY written
// in place, e.g. a TLS task of the multi-rank stealing scheme: every writer of
// address a offers (gid+1) << 32 | (current value of a), so the max is the last
// writer's key carrying the final value (reading A9).  Keys only for the arrays
// that have a key table (indirect writes); identity outputs stay where they are.
template <int OP, int DT>
__global__ void __launch_bounds__(256) k_export_keys(DLoop L, unsigned long long *kA, unsigned long long *kT) {
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < L.n; i += stride) {
    if (kA) {
      const int64_t a = ixl(L, L.w, i);
      atomicMax(&kA[a], pack_key(L.base + i, __ldcg(L.A + a)));
    }
    if constexpr (OP == JP_OP_PRIV_TMP) {
      if (kT) {
        const int64_t b = ixl(L, L.s, i);
        atomicMax(&kT[b], pack_key(L.base + i, __ldcg(L.T + b)));
      }
    }
  }
}

template <int OP, int DT>
static void run_export(const DLoop &d, unsigned long long *kA, unsigned long long *kT, cudaStream_t st) {
  int64_t need = (d.n + 255) / 256, cap = (int64_t)num_sms() * 8;
  k_export_keys<OP, DT><<<(int)(need < cap ? need : cap), 256, 0, st>>>(d, kA, kT);
  note_launch();
}

cudaError_t launch_export_keys(const Job &j, void *ws, const Layout &lo, cudaStream_t st) {
  if (j.d.n == 0) return cudaSuccess;
  JP_DISPATCH(j.op, j.dt, run_export, j.d, at<unsigned long long>(ws, lo, R_KEYS_A),
              at<unsigned long long>(ws, lo, R_KEYS_T), st);
  return launch_check();
}

// ---------------------------------------------------------------------------
// Task stealing on the device (Alg. 1: "steal when empty"): the
// privatized body over a list of chunks dealt to the ranks, each rank's block
// claimed ascending by its owner and descending by idle ranks through one
// system-scope atomicAdd on a packed (tail << 32 | head) counter per rank
// (the same protocol as k_doall_spill).  Every rank works on its own replica:
// exposed reads see the replica (legal: d_raw = 0 for these chunks), keyed
// writes go to the rank's key tables (merged afterwards by C4), identity
// writes are stored in place (unique per iteration).
// ---------------------------------------------------------------------------
constexpr int kClaimRanks = 8;
struct ClaimArgs {
  DLoop L;
  const int64_t *chunks;            // [2 * nchunks] local (start, end)
  int64_t first[kClaimRanks + 1];   // rank k owns chunk entries [first[k], first[k+1])
  unsigned long long *ctr, *kA, *kT;
  int64_t *stats;                   // [0] own iterations, [1] stolen iterations, [2] stolen chunks
  int world, me;
};

__device__ __forceinline__ bool claim_chunk(unsigned long long *ctr, int64_t nb, bool tail, int64_t &c) {
  const unsigned long long old = atomicAdd_system(ctr, tail ? (1ull << 32) : 1ull);
  const int64_t h = (uint32_t)old, t = (uint32_t)(old >> 32);
  if (h + t >= nb) return false;
  c = tail ? nb - 1 - t : h;
  return true;
}

template <int OP, int DT>
__global__ void __launch_bounds__(256) k_priv_claim(const __grid_constant__ ClaimArgs P) {
  __shared__ int s_rank;
  __shared__ long long s_idx;
  const DLoop &L = P.L;
  int64_t own = 0, stolen = 0, nst = 0;
  bool mine = true;
  for (;;) {
    if (threadIdx.x == 0) {
      int rk = -1;
      int64_t c = 0;
      const int64_t nbm = P.first[P.me + 1] - P.first[P.me];
      if (mine && claim_chunk(&P.ctr[P.me], nbm, false, c)) rk = P.me;
      else mine = false;
      while (rk < 0) {   // the rank with the most unclaimed chunks, ties to the lowest
        int best = -1;
        int64_t most = 0;
        for (int k = 0; k < P.world; k++) {
          if (k == P.me) continue;
          const unsigned long long v = *(volatile unsigned long long *)&P.ctr[k];
          const int64_t left = P.first[k + 1] - P.first[k] - (int64_t)(uint32_t)v - (int64_t)(uint32_t)(v >> 32);
          if (left > most) { most = left; best = k; }
        }
        if (best < 0) break;
        if (claim_chunk(&P.ctr[best], P.first[best + 1] - P.first[best], true, c)) rk = best;
      }
      s_rank = rk;
      s_idx = rk < 0 ? 0 : P.first[rk] + c;
    }
    __syncthreads();
    const int rk = s_rank;
    const int64_t ci = s_idx;
    __syncthreads();
    if (rk < 0) break;
    const int64_t cs = P.chunks[2 * ci], ce = P.chunks[2 * ci + 1];
    for (int64_t i = cs + threadIdx.x; i < ce; i += blockDim.x) {
      uint32_t va = 0, vt = 0;
      body_values<OP, DT>(L, i, L.A, va, vt);
      const int64_t a = ixl(L, L.w, i);
      if (P.kA) atomicMax(&P.kA[a], pack_key(L.base + i, va));
      else L.A[a] = va;
      if constexpr (OP == JP_OP_PRIV_TMP) {
        const int64_t b = ixl(L, L.s, i);
        if (P.kT) atomicMax(&P.kT[b], pack_key(L.base + i, vt));
        else L.T[b] = vt;
      }
    }
    if (threadIdx.x == 0) {
      if (rk == P.me) own += ce - cs;
      else { stolen += ce - cs; nst++; }
    }
  }
  if (threadIdx.x == 0 && P.stats) {
    if (own) atomicAdd(reinterpret_cast<unsigned long long *>(&P.stats[0]), (unsigned long long)own);
    if (stolen) {
      atomicAdd(reinterpret_cast<unsigned long long *>(&P.stats[1]), (unsigned long long)stolen);
      atomicAdd(reinterpret_cast<unsigned long long *>(&P.stats[2]), (unsigned long long)nst);
    }
  }
}

template <int OP, int DT>
static void run_claim(const ClaimArgs &P, int grid, cudaStream_t st) {
  k_priv_claim<OP, DT><<<grid, 256, 0, st>>>(P);
  note_launch();
}

cudaError_t launch_priv_claim(const Job &j, void *ws, const Layout &lo, const int64_t *chunks, const int64_t *first,
                              int world, int me, unsigned long long *ctr, int64_t *stats, int max_ctas,
                              cudaStream_t st) {
  ClaimArgs P;
  memset(&P, 0, sizeof P);
  P.L = j.d;
  P.chunks = chunks;
  for (int k = 0; k <= world; k++) P.first[k] = first[k];
  P.ctr = ctr;
  P.kA = at<unsigned long long>(ws, lo, R_KEYS_A);
  P.kT = j.op == JP_OP_PRIV_TMP ? at<unsigned long long>(ws, lo, R_KEYS_T) : nullptr;
  P.stats = stats;
  P.world = world;
  P.me = me;
  int grid = num_sms() * 4;
  if (max_ctas > 0 && grid > max_ctas) grid = max_ctas;
  JP_DISPATCH(j.op, j.dt, run_claim, P, grid, st);
  return launch_check();
}

// ---------------------------------------------------------------------------
// C4 over NVLink peer memory (SURVEY §2c C9's role, without NCCL): one CTA per
// rank reads every rank's key table (CUDA-IPC-mapped device pointers), keeps
// the maximum per slot and applies it.  Two device-side barriers on a
// monotone counter in rank 0's memory (system-scope atomics, acquire loads)
// bracket the reads: every rank's keys are in before anyone reads (phase A),
// and nobody clears its table for the next call before every rank has read it
// (phase B).  epoch = 1, 2, ... per call; the counter is never reset.
// A wait longer than ~4 s sets *err and abandons the merge (no hang).
// ---------------------------------------------------------------------------
constexpr int kMaxPeers = 8;
struct PeerKeys {
  const unsigned long long *k[kMaxPeers];
};

__device__ __forceinline__ unsigned long long ld_acquire_sys(const unsigned long long *p) {
  unsigned long long v;
  asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ unsigned long long ld_relaxed_sys(const unsigned long long *p) {
  unsigned long long v;
  asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ unsigned long long gtimer() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
__device__ bool p2p_barrier(unsigned long long *bar, unsigned long long target, int *err) {
  __shared__ int ok;
  if (threadIdx.x == 0) {
    __threadfence_system();
    atomicAdd_system(bar, 1ull);
    const unsigned long long t0 = gtimer();
    ok = 1;
    while (ld_acquire_sys(bar) < target) {
      if (gtimer() - t0 > 4000000000ull) { ok = 0; atomicExch(err, 1); break; }
      __nanosleep(200);
    }
  }
  __syncthreads();
  return ok;
}

__global__ void __launch_bounds__(1024) k_keys_merge_p2p(PeerKeys P, int world, unsigned long long *mine, int64_t len,
                                                         unsigned long long *bar, unsigned long long epoch,
                                                         uint32_t *arr, int *err) {
  extern __shared__ unsigned long long mx[];   // len <= kP2PMaxLen
  if (!p2p_barrier(bar, (2 * epoch - 1) * (unsigned long long)world, err)) return;
  for (int64_t a = threadIdx.x; a < len; a += blockDim.x) {
    unsigned long long m = 0;
    for (int k = 0; k < world; k++) {
      const unsigned long long v = ld_relaxed_sys(P.k[k] + a);
      m = v > m ? v : m;
    }
    mx[a] = m;
  }
  __syncthreads();
  if (!p2p_barrier(bar, 2 * epoch * (unsigned long long)world, err)) return;
  for (int64_t a = threadIdx.x; a < len; a += blockDim.x) {
    const unsigned long long m = mx[a];
    mine[a] = m;
    if (arr && m) arr[a] = (uint32_t)m;
  }
}

cudaError_t launch_keys_merge_p2p(const unsigned long long *const *peers, int world, unsigned long long *mine,
                                  int64_t len, unsigned long long *bar, unsigned long long epoch, uint32_t *arr,
                                  int *err, cudaStream_t st) {
  PeerKeys P;
  for (int k = 0; k < kMaxPeers; k++) P.k[k] = k < world ? peers[k] : nullptr;
  const size_t smem = 8 * (size_t)(len > 0 ? len : 1);
  if (smem > 48 * 1024) set_smem_once((const void *)k_keys_merge_p2p, (int)smem);
  k_keys_merge_p2p<<<1, 1024, smem, st>>>(P, world, mine, len, bar, epoch, arr, err);
  note_launch();
  return launch_check();
}

cudaError_t launch_merge_apply(void *arr, int64_t len, const int64_t *keys, cudaStream_t st) {
  apply(static_cast<uint32_t *>(arr), len, reinterpret_cast<const unsigned long long *>(keys), st);
  return launch_check();
}

}  // namespace jp

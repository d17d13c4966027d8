// jp_internal.cuh -- device-side helpers of libjp.so (product path only).
//
// Nothing here is shared with oracle/: the loop bodies, access sets and
// encodings below are re-derived from the paper and DESIGN.md, not included
// from the oracle (task rule: the two sides share no code).
#pragma once
#include <cstdint>
#include <cuda_runtime.h>
#include "../../include/jp.h"

// CTA-wide barrier used by every kernel of the library: an explicit
// barrier.sync with a memory clobber (see jp_tls.cu TLS_SYNC and DESIGN.md
// Sec.6 for the intermittent failure observed with __syncthreads()).
#define JP_CTA_SYNC() asm volatile("barrier.sync 0;" ::: "memory")

namespace jp {

constexpr int kSmemSlots = 4096;          // arrays this small are pre-aggregated per CTA
#ifndef JP_TLS_THREADS
#define JP_TLS_THREADS 512
#endif
#ifndef JP_TLS_IPT
#define JP_TLS_IPT 8
#endif
#ifndef JP_TLS_HASHLOG
#define JP_TLS_HASHLOG 13
#endif
constexpr int kTlsCtaThreads = JP_TLS_THREADS;   // single-CTA TLS path
constexpr int kTlsCtaIpt = JP_TLS_IPT;           // -> W <= 4096
constexpr int kTlsCtaWmax = kTlsCtaThreads * kTlsCtaIpt;
constexpr int kTlsFillThreads = 128;             // threads that issue the index-ring copies
constexpr int kTlsHashLog = JP_TLS_HASHLOG;      // 8192 slots = 2 x W_max
constexpr int kTlsHash = 1 << kTlsHashLog;
constexpr int kTlsGridThreads = 512;
constexpr uint32_t kEmpty = 0xFFFFFFFFu;

// Header slots (int64) at the start of every workspace.
enum Hdr : int {
  H_RAW = 0, H_WAR = 1, H_WAW = 2, H_FIRST_RAW = 3, H_BAD = 4,
  H_TLS_COMMITTED = 8, H_TLS_EXECUTED = 9, H_TLS_WINDOWS = 10, H_TLS_VIOL = 11, H_TINY_MODE = 12,
  H_TINY_WMAX = 13, H_TINY_REC = 14,
  H_BAR_COUNT = 16, H_BAR_GEN = 17, H_FV0 = 20, H_FV1 = 21, H_FV2 = 22, H_AFFINE = 24 /* 2 slots = 4 int */,
  H_PRED_FAIL = 28 /* buckets whose writers overflowed the last-writer pass (jp_bucket.cu) */,
  H_PRED_SEG = 29 /* longest writer list of one address seen by that pass */,
  H_GATE = 30 /* nonzero: the index arrays look affine on their prefix -- the profile's kernels exit */,
  H_DIST = 64 /* 32 slots: raw reads by floor(log2(i - writer)) */, H_SLOTS = 96
};
constexpr size_t kHeaderBytes = 4096;

// The loop as seen by kernels: element arrays are 32-bit words, the dtype is a
// template parameter of every kernel.
struct DLoop {
  int64_t n, base;
  int64_t ioff;              // identity index of local iteration i is ioff + i (sub-loops)
  const int32_t *r, *r2, *w, *s;
  uint32_t *A; int64_t lenA;
  const uint32_t *X; int64_t lenX;
  uint32_t *T; int64_t lenT;
  uint32_t c0, c1;
  // nullable device flag (the index-validation count): kernels of a run that
  // was launched before its validation result is known exit at once when it is
  // nonzero, so an out-of-range index still leaves every array untouched (A13)
  const int64_t *abort = nullptr;
};

__device__ __forceinline__ bool aborted(const DLoop &L) {
  return L.abort && *reinterpret_cast<const volatile int64_t *>(L.abort) != 0;
}

// index of local iteration i through index array p (NULL => identity)
__host__ __device__ inline int64_t ixl(const DLoop &L, const int32_t *p, int64_t i) {
  return p ? (int64_t)p[i] : L.ioff + i;
}

// --- fp32 / int32 arithmetic: one IEEE RN op per operator, never contracted
// (reading A12), or two's-complement wrap (reading A11).
template <int DT> __device__ __forceinline__ uint32_t op_add(uint32_t a, uint32_t b) {
  if constexpr (DT == JP_I32) return a + b;
  else return __float_as_uint(__fadd_rn(__uint_as_float(a), __uint_as_float(b)));
}
template <int DT> __device__ __forceinline__ uint32_t op_mul(uint32_t a, uint32_t b) {
  if constexpr (DT == JP_I32) return a * b;
  else return __float_as_uint(__fmul_rn(__uint_as_float(a), __uint_as_float(b)));
}

// Which arrays can carry a cross-iteration conflict: an array reached through
// at least one non-identity index (otherwise iteration i only touches element i).
__host__ __device__ inline bool a_indirect(int op, const int32_t *r, const int32_t *r2, const int32_t *w) {
  switch (op) {
    case JP_OP_ADD_C: return r || w;
    case JP_OP_SAXPY: return w != nullptr;          // Y read and written through w
    case JP_OP_PRIV_TMP: return w != nullptr;       // Y only written
    default: return r || r2 || w;                   // STENCIL2
  }
}
__host__ __device__ inline bool a_has_reads(int op) { return op != JP_OP_PRIV_TMP; }
__host__ __device__ inline bool t_indirect(int op, const int32_t *s) { return op == JP_OP_PRIV_TMP && s; }

// Exposed-read encoding of the profile tables: INT32_MAX - gid, empty -1, so
// that max == earliest; "some earlier iteration touched a" <=> tab[a] > enc(i).
__device__ __forceinline__ int32_t enc_gid(int64_t gid) { return (int32_t)(0x7FFFFFFF - gid); }

// Packed last-writer key: (gid+1) << 32 | bits(value); empty 0 (reading A9).
__device__ __forceinline__ unsigned long long pack_key(int64_t gid, uint32_t v) {
  return ((unsigned long long)(gid + 1) << 32) | v;
}

// Values the body of iteration i writes, computed from `src` reads.
// PRIV_TMP: vt is the private T value, va the Y value.
template <int OP, int DT>
__device__ __forceinline__ void body_values(const DLoop &L, int64_t i, const uint32_t *srcA,
                                            uint32_t &va, uint32_t &vt) {
  if constexpr (OP == JP_OP_ADD_C) {
    va = op_add<DT>(srcA[ixl(L, L.r, i)], L.c0);
  } else if constexpr (OP == JP_OP_SAXPY) {
    va = op_add<DT>(op_mul<DT>(L.c0, L.X[ixl(L, L.r, i)]), srcA[ixl(L, L.w, i)]);
  } else if constexpr (OP == JP_OP_PRIV_TMP) {
    vt = op_mul<DT>(L.c0, L.X[ixl(L, L.r, i)]);
    va = op_add<DT>(vt, L.c1);
  } else {
    va = op_mul<DT>(op_add<DT>(srcA[ixl(L, L.r, i)], srcA[ixl(L, L.r2, i)]), L.c0);
  }
}

// --- bulk-copy (TMA 1-D) + mbarrier helpers (sm_90+ PTX), used by the staged stream kernels
__device__ __forceinline__ uint32_t smem_u32(const void *p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void mbar_init(unsigned long long *b, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(b)), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_expect_tx(unsigned long long *b, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(b)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void mbar_wait(unsigned long long *b, uint32_t parity) {
  asm volatile(
      "{\n\t.reg .pred p;\n"
      "WAIT_%=:\n\t"
      "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t"
      "@!p bra WAIT_%=;\n\t}" ::"r"(smem_u32(b)), "r"(parity) : "memory");
}
__device__ __forceinline__ void bulk_load(void *dst, const void *src, uint32_t bytes, unsigned long long *bar) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
               ::"r"(smem_u32(dst)), "l"(src), "r"(bytes), "r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ void bulk_store(void *dst, const void *src, uint32_t bytes) {
  asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst), "r"(smem_u32(src)), "r"(bytes)
               : "memory");
}

// Launch bookkeeping (counted for bench.py's gpu_launches).
void note_launch(int k = 1);
int num_sms();
cudaError_t launch_check();

}  // namespace jp

// op x dtype dispatch to a templated functor call
#define JP_DISPATCH(OPV, DTV, FN, ...)                                             \
  do {                                                                             \
    switch ((OPV) * 2 + (DTV)) {                                                   \
      case 0: FN<JP_OP_ADD_C, JP_I32>(__VA_ARGS__); break;                         \
      case 1: FN<JP_OP_ADD_C, JP_F32>(__VA_ARGS__); break;                         \
      case 2: FN<JP_OP_SAXPY, JP_I32>(__VA_ARGS__); break;                         \
      case 3: FN<JP_OP_SAXPY, JP_F32>(__VA_ARGS__); break;                         \
      case 4: FN<JP_OP_PRIV_TMP, JP_I32>(__VA_ARGS__); break;                      \
      case 5: FN<JP_OP_PRIV_TMP, JP_F32>(__VA_ARGS__); break;                      \
      case 6: FN<JP_OP_STENCIL2, JP_I32>(__VA_ARGS__); break;                      \
      case 7: FN<JP_OP_STENCIL2, JP_F32>(__VA_ARGS__); break;                      \
    }                                                                              \
  } while (0)

/*
 * oracle/jpo.h -- TEST INFRASTRUCTURE ONLY.  This is NOT the product path.
 *
 * A plain, slow, sequential CPU oracle for the Japonica loop-mode hot path
 * (Han, Zhang, Lam, Wang, ICPP'13; /root/reference/PAPER.md, cited "P:L<n>").
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / reference
 * leg may load it.  It shares NO code, header, table or constant with the CUDA
 * library (paper_conf_icpp_hanzlw13_b200/csrc, include/jp.h); every type below
 * is declared independently on purpose.
 *
 * Loop model (SURVEY.md Sec.8 "Body opcodes"): one annotated
 * `for (i = 0; i < n; i++)` loop (Table I) whose body is
 * one of four fixed opcodes over int32 or fp32 element arrays, indexed through
 * int32 index arrays (NULL => identity i):
 *   ADD_C    A[w[i]] = A[r[i]] + c0
 *   SAXPY    Y[w[i]] = c0*X[r[i]] + Y[w[i]]          (Y lives in the A slot)
 *   PRIV_TMP T[s[i]] = c0*X[r[i]]; Y[w[i]] = T[s[i]] + c1   (T = private(list))
 *   STENCIL2 A[w[i]] = (A[r[i]] + A[r2[i]]) * c0      (Gauss-Seidel shape)
 * int32 arithmetic wraps (reading A11: Java int); fp32 arithmetic is one IEEE
 * round-to-nearest-even operation per C operator, no contraction, no FTZ
 * (reading A12: Java float) -- this file MUST be compiled with
 * -ffp-contract=off and without -ffast-math.
 */
#ifndef JPO_ORACLE_H
#define JPO_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

enum { JPO_OP_ADD_C = 0, JPO_OP_SAXPY = 1, JPO_OP_PRIV_TMP = 2, JPO_OP_STENCIL2 = 3 };
enum { JPO_I32 = 0, JPO_F32 = 1 };
enum { JPO_OK = 0, JPO_ERR_ARG = -1, JPO_ERR_INDEX = -5 };
/* array ids used in access lists */
enum { JPO_ARR_A = 0, JPO_ARR_X = 1, JPO_ARR_T = 2 };

typedef struct {
  int64_t n;                 /* trip count                                  */
  int32_t op, dtype;         /* JPO_OP_*, JPO_I32/JPO_F32                   */
  const int32_t *r, *r2, *w, *s;   /* NULL => identity i                    */
  void *A; int64_t len_A;    /* ADD_C/STENCIL2: A;  SAXPY/PRIV_TMP: Y       */
  const void *X; int64_t len_X;
  void *T; int64_t len_T;
  uint32_t c0, c1;           /* raw 32-bit patterns of the constants        */
} jpo_loop;

typedef struct {
  int64_t n, raw_iters, war_iters, waw_iters, first_raw_iter;
  int64_t raw_pairs, war_pairs, waw_pairs;   /* jpo_pairs only; -1 otherwise */
} jpo_profile;

typedef struct { int64_t committed, executed, windows, violations; } jpo_tls_stats;

/* Sequential definition. Index check first; on any
 * out-of-range index nothing is modified and JPO_ERR_INDEX is returned (A13). */
int jpo_run_seq(const jpo_loop *L);
/* Same body, executed in the order given by perm[0..n) (DOALL-legality pin). */
int jpo_run_order(const jpo_loop *L, const int64_t *perm);
/* Single ascending pass with first-writer / read-before maps (item 2).
 * flags (nullable, uint8[n]): bit0 raw_i, bit1 war_i, bit2 waw_i.          */
int jpo_profile_run(const jpo_loop *L, jpo_profile *out, uint8_t *flags);
/* O(n^2) enumeration of all ordered pairs (item 3); same flags + pair counts. */
int jpo_pairs(const jpo_loop *L, jpo_profile *out, uint8_t *flags);
/* RAW sources: src[j] = 1 iff a write of j is exposed-read by some i > j. */
int jpo_raw_sources(const jpo_loop *L, uint8_t *src);
/* Windowed TLS as a definition (item 4).  window > 0: fixed W.  window == 0:
 * adaptive policy of reading A8 with cap w_max; prof_raw_iters < 0 means "no
 * profile known".  Modifies the arrays (must end equal to jpo_run_seq).      */
int jpo_sim_tls(const jpo_loop *L, int64_t window, int64_t w_max,
                int64_t prof_raw_iters, jpo_tls_stats *st);
/* The adaptive window policy of reading A8, exposed for pinning.
 * prev_commit < 0 => initial window.                                         */
int64_t jpo_tls_next_window(int64_t n, int64_t prof_raw_iters, int64_t prev_commit,
                            int64_t w_max);
/* Windowed TLS with on-chip recovery (reading B7):
 * fixed windows [kW, (k+1)W).  In each window every iteration speculates
 * against the memory of the window start (SE); DC marks the iterations with an
 * exposed read written by an EARLIER iteration of the same window ("which
 * threads fell in violation"); the non-violators commit and the
 * violators are recovered, so the window ends in the sequential state.
 * stats: windows; violations = violating iterations (each re-executed once);
 * executed = n + violations; committed = n.  window > 0.                    */
int jpo_sim_tls_fwd(const jpo_loop *L, int64_t window, jpo_tls_stats *st);
/* Privatized semantics (item 5 / readings A9, A10). */
int jpo_sim_priv(const jpo_loop *L);

#ifdef __cplusplus
}
#endif
#endif

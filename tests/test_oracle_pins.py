"""Pins of the CPU oracle against things other than itself (-m "not gpu").

Each pin is chosen so that a plausible mistake in oracle/jpo.c (a dropped
access, a swapped r/w, a wrong window bound, FMA contraction, a missed WAR on a
covered read) fails at least one of them:
  * hand-worked N=8 tables (tests/golden/addc_n8.txt),
  * closed forms (permutation self-update, prefix chain, read-ahead shift,
    Gauss-Seidel STENCIL2, PRIV_TMP last-writer),
  * a pure-Python brute force over all ordered pairs, written here from the
    definition (reading A1), exhaustive over all (r, w) in [0,3)^5,
  * a pure-Python O(W^2) TLS window simulator (reading A6) on small loops,
  * exact-rational IEEE rounding for the fp32 bodies (reading A12),
  * invariants (d = 0 => zero violations, ...).
"""
import fractions
import itertools
import os

import numpy as np
import pytest

import oracle as O

OPS = {"ADD_C": O.OP_ADD_C, "SAXPY": O.OP_SAXPY, "PRIV_TMP": O.OP_PRIV_TMP, "STENCIL2": O.OP_STENCIL2}


# ----------------------------------------------------------------------------
# independent restatement of the access sets (SURVEY Sec.8 opcode table)
# ----------------------------------------------------------------------------
def acc_sets(op, i, r, r2, w, s):
    ix = lambda a: i if a is None else int(a[i])  # noqa: E731
    if op == O.OP_ADD_C:
        return [("A", ix(r))], [], [("A", ix(w))]
    if op == O.OP_SAXPY:
        return [("X", ix(r)), ("A", ix(w))], [], [("A", ix(w))]
    if op == O.OP_PRIV_TMP:
        return [("X", ix(r))], [("T", ix(s))], [("T", ix(s)), ("A", ix(w))]
    return [("A", ix(r)), ("A", ix(r2))], [], [("A", ix(w))]


def brute_profile(op, n, r=None, r2=None, w=None, s=None):
    """Reading A1 written out over all ordered pairs j < i."""
    sets = [acc_sets(op, i, r, r2, w, s) for i in range(n)]
    raw = war = waw = 0
    flags = []
    for i in range(n):
        rexp_i, _, w_i = sets[i]
        f_raw = any(set(sets[j][2]) & set(rexp_i) for j in range(i))
        f_war = any(set(sets[j][0] + sets[j][1]) & set(w_i) for j in range(i))
        f_waw = any(set(sets[j][2]) & set(w_i) for j in range(i))
        raw += f_raw; war += f_war; waw += f_waw
        flags.append(int(f_raw) | int(f_war) << 1 | int(f_waw) << 2)
    return raw, war, waw, flags


def brute_sources(op, n, r=None, r2=None, w=None, s=None):
    """RAW sources over all ordered pairs: j with W(j) ∩ R_exp(i) != {} for an i > j."""
    sets = [acc_sets(op, i, r, r2, w, s) for i in range(n)]
    return [int(any(set(sets[j][2]) & set(sets[i][0]) for i in range(j + 1, n))) for j in range(n)]


def brute_tls_stats(op, n, W, r=None, r2=None, w=None, s=None):
    """Reading A6: fv = first i in the window with an earlier in-window writer of
    one of its exposed reads (O(W^2)); prefix commit; restart at fv."""
    sets = [acc_sets(op, i, r, r2, w, s) for i in range(n)]
    ws, windows, viol, executed = 0, 0, 0, 0
    while ws < n:
        we = min(ws + W, n)
        fv = we
        for i in range(ws, we):
            if any(set(sets[j][2]) & set(sets[i][0]) for j in range(ws, i)):
                fv = i
                break
        windows += 1
        viol += fv < we
        executed += we - ws
        ws = fv
    return {"committed": n, "executed": executed, "windows": windows, "violations": viol}


def _arr(tok):
    return None if tok.strip() == "-" else np.array([int(t) for t in tok.split()], dtype=np.int32)


def load_golden(golden_dir):
    rows = []
    with open(os.path.join(golden_dir, "addc_n8.txt")) as f:
        for line in f:
            if line.startswith("#") or not line.strip():
                continue
            p = [t.strip() for t in line.split("|")]
            rows.append(dict(name=p[0], op=OPS[p[1]], c0=int(p[2]), A0=_arr(p[3]), r=_arr(p[4]), r2=_arr(p[5]),
                             w=_arr(p[6]), A=_arr(p[7]), prof=[int(t) for t in p[8].split()],
                             tls=[int(t) for t in p[9].split()]))
    return rows


# ----------------------------------------------------------------------------
def test_golden_tables(golden_dir):
    for g in load_golden(golden_dir):
        L = O.Loop(g["op"], O.I32, 8, g["A0"], r=g["r"], r2=g["r2"], w=g["w"], c0=g["c0"])
        st, A, _ = O.run_seq(L)
        assert st == O.OK
        assert A.tolist() == g["A"].tolist(), g["name"]
        p = O.profile(L)
        assert [p["raw_iters"], p["war_iters"], p["waw_iters"]] == g["prof"], g["name"]
        W, windows, viol, executed = g["tls"]
        st, A2, _, stats = O.sim_tls(L, W)
        assert A2.tolist() == g["A"].tolist(), g["name"]
        assert (stats["windows"], stats["violations"], stats["executed"], stats["committed"]) == (windows, viol, executed, 8)


@pytest.mark.parametrize("n", [1, 2, 7, 64, 1000])
def test_closed_forms_addc(n):
    rng = np.random.default_rng(n)
    A0 = rng.integers(-2**31, 2**31, size=n, dtype=np.int64).astype(np.int32)
    c = 2**31 - 5  # forces int32 wrap
    u = A0.astype(np.uint32)
    # permutation self-update r = w = pi: A'[a] = A[a] + c
    pi = rng.permutation(n).astype(np.int32)
    L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=pi, w=pi, c0=c)
    assert O.run_seq(L)[1].view(np.uint32).tolist() == ((u + np.uint32(c)) & 0xFFFFFFFF).tolist()
    p = O.profile(L)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (0, 0, 0)
    # prefix chain: A'[i] = A[0] + (i+1) c  (mod 2^32)
    L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=np.maximum(np.arange(n) - 1, 0), w=np.arange(n), c0=c)
    exp = [(int(u[0]) + (i + 1) * c) & 0xFFFFFFFF for i in range(n)]
    assert O.run_seq(L)[1].view(np.uint32).tolist() == exp
    p = O.profile(L)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (max(n - 1, 0), 0, 0)
    assert p["first_raw_iter"] == (1 if n > 1 else -1)
    _, _, _, st = O.sim_tls(L, 4)
    if n > 1:
        assert (st["windows"], st["violations"]) == (n, n - 1)
    # read-ahead shift: pure WAR
    r = np.minimum(np.arange(n) + 1, n - 1)
    L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=r, w=np.arange(n), c0=c)
    exp = [(int(u[min(i + 1, n - 1)]) + c) & 0xFFFFFFFF for i in range(n)]
    assert O.run_seq(L)[1].view(np.uint32).tolist() == exp
    p = O.profile(L)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (0, max(n - 1, 0), 0)
    # Gauss-Seidel STENCIL2: (N-1, N-1, 0)
    L = O.Loop(O.OP_STENCIL2, O.I32, n, A0, r=np.maximum(np.arange(n) - 1, 0), r2=np.minimum(np.arange(n) + 1, n - 1),
               w=np.arange(n), c0=3)
    p = O.profile(L)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (max(n - 1, 0), max(n - 1, 0), 0)


def test_profile_exhaustive_vs_bruteforce():
    """All ADD_C loops with N=5 over |A|=3: (r, w) in [0,3)^5 x [0,3)^5 (59049 loops)."""
    n, la = 5, 3
    A0 = np.array([5, -3, 11], dtype=np.int32)
    seen_zero = 0
    for rw in itertools.product(range(la), repeat=2 * n):
        r = np.array(rw[:n], dtype=np.int32)
        w = np.array(rw[n:], dtype=np.int32)
        L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=r, w=w, c0=7)
        p = O.profile(L)
        b = brute_profile(O.OP_ADD_C, n, r=r, w=w)
        assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == b[:3]
        assert p["flags"].tolist() == b[3]
        assert O.raw_sources(L).tolist() == brute_sources(O.OP_ADD_C, n, r=r, w=w)
        if p["raw_iters"] == 0:
            seen_zero += 1
    assert seen_zero == 1728  # the count the survey's brute force found


@pytest.mark.parametrize("seed", range(40))
def test_profile_random_all_ops_vs_bruteforce(seed):
    rng = np.random.default_rng(100 + seed)
    n = int(rng.integers(1, 17))
    op = seed % 4
    la, lx, lt = int(rng.integers(1, 6)), int(rng.integers(n, n + 4)), int(rng.integers(1, 5))
    mk = lambda hi: rng.integers(0, hi, size=n).astype(np.int32) if rng.random() < 0.8 else None  # noqa: E731
    r = mk(lx if op in (O.OP_SAXPY, O.OP_PRIV_TMP) else la)
    if op in (O.OP_SAXPY, O.OP_PRIV_TMP) and r is None and lx < n:
        lx = n
    w = mk(la)
    if w is None:
        la = max(la, n)
    if op in (O.OP_ADD_C, O.OP_STENCIL2) and r is None:
        la = max(la, n)
    r2 = mk(la) if op == O.OP_STENCIL2 else None
    if op == O.OP_STENCIL2 and r2 is None:
        la = max(la, n)
    s = rng.integers(0, lt, size=n).astype(np.int32) if op == O.OP_PRIV_TMP else None
    dt = O.F32 if seed % 3 == 0 else O.I32
    el = np.float32 if dt == O.F32 else np.int32
    L = O.Loop(op, dt, n, rng.integers(-9, 9, size=la).astype(el), r=r, r2=r2, w=w, s=s,
               X=rng.integers(-9, 9, size=lx).astype(el), T=rng.integers(-9, 9, size=lt).astype(el), c0=3, c1=1)
    p, q = O.profile(L), O.pairs(L)
    b = brute_profile(op, n, r=r, r2=r2, w=w, s=s)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == b[:3]
    assert p["flags"].tolist() == b[3] == q["flags"].tolist()
    assert O.raw_sources(L).tolist() == brute_sources(op, n, r=r, r2=r2, w=w, s=s)
    # TLS: arrays equal the sequential run, stats equal the O(W^2) definition
    for W in (1, 2, 3, 5, 16):
        st, A, T, stats = O.sim_tls(L, W)
        _, A0, T0 = O.run_seq(L)
        assert A.tobytes() == A0.tobytes() and (T is None or T.tobytes() == T0.tobytes())
        assert stats == brute_tls_stats(op, n, W, r=r, r2=r2, w=w, s=s)
        assert stats["violations"] <= p["raw_iters"]


def test_tls_exhaustive_invariants():
    """N=5, |A|=3, every (r, w), W in {1,2,3,5}: TLS == sequential; d_raw = 0 =>
    0 violations and ceil(N/W) windows; privatized == sequential iff allowed."""
    n, la = 5, 3
    A0 = np.array([5, -3, 11], dtype=np.int32)
    for rw in itertools.product(range(la), repeat=2 * n):
        r = np.array(rw[:n], dtype=np.int32)
        w = np.array(rw[n:], dtype=np.int32)
        L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=r, w=w, c0=7)
        seq = O.run_seq(L)[1]
        raw = O.profile(L)["raw_iters"]
        for W in (1, 2, 3, 5):
            _, A, _, st = O.sim_tls(L, W)
            assert A.tolist() == seq.tolist()
            assert st["committed"] == n and st["violations"] <= raw
            if raw == 0:
                assert st["violations"] == 0 and st["windows"] == -(-n // W)
        if raw == 0:
            assert O.sim_priv(L)[1].tolist() == seq.tolist()


@pytest.mark.parametrize("n", [1, 2, 9, 500])
def test_raw_sources_closed_forms(n):
    """Closed forms: the prefix chain's sources are every iteration but the last;
    a permutation self-update has none; Gauss-Seidel's are all but the last."""
    ar = np.arange(n, dtype=np.int32)
    A0 = np.zeros(n, dtype=np.int32)
    pc = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=np.maximum(ar - 1, 0), w=ar, c0=1)
    # j writes j and iteration j+1 reads it; the last write is never read later
    assert O.raw_sources(pc).tolist() == [1] * (n - 1) + [0]
    perm = np.random.default_rng(n).permutation(n).astype(np.int32)
    assert O.raw_sources(O.Loop(O.OP_ADD_C, O.I32, n, A0, r=perm, w=perm, c0=1)).tolist() == [0] * n
    gs = O.Loop(O.OP_STENCIL2, O.I32, n, A0, r=np.maximum(ar - 1, 0), r2=np.minimum(ar + 1, n - 1), w=ar, c0=1)
    # j is read later by j+1 (through r = j); the last iteration's write is never read later
    assert O.raw_sources(gs).tolist() == [1] * (n - 1) + [0]


def test_priv_counterexample_prefix_chain():
    """RAW forbids privatization: on the prefix chain privatized != sequential."""
    n = 8
    L = O.Loop(O.OP_ADD_C, O.I32, n, np.arange(n) * 10, r=np.maximum(np.arange(n) - 1, 0), w=np.arange(n), c0=7)
    assert O.sim_priv(L)[1].tolist() != O.run_seq(L)[1].tolist()


# ----------------------------------------------------------------------------
# fp32: exact-rational IEEE round-to-nearest-even (reading A12)
# ----------------------------------------------------------------------------
def rn32(q: fractions.Fraction) -> np.float32:
    """Round an exact rational to the nearest fp32 (ties to even); normal range only."""
    if q == 0:
        return np.float32(0.0)
    sign = -1 if q < 0 else 1
    q = abs(q)
    e = q.numerator.bit_length() - q.denominator.bit_length()
    while fractions.Fraction(2) ** e > q:
        e -= 1
    while fractions.Fraction(2) ** (e + 1) <= q:
        e += 1
    ulp = fractions.Fraction(2) ** (e - 23)
    m = q / ulp
    fl = m.numerator // m.denominator
    rem = m - fl
    if rem > fractions.Fraction(1, 2) or (rem == fractions.Fraction(1, 2) and fl % 2 == 1):
        fl += 1
    return np.float32(sign * float(fl * ulp))


F = lambda x: fractions.Fraction(float(x))  # noqa: E731


def test_fp32_saxpy_two_roundings():
    """SAXPY must be fl(fl(c0*x) + y), never the fused fl(c0*x + y)."""
    rng = np.random.default_rng(7)
    n = 4096
    X = ((rng.integers(0, 2**23, size=n) * 2.0**-22) - 1).astype(np.float32)
    Y = ((rng.integers(0, 2**23, size=n) * 2.0**-22) - 1).astype(np.float32)
    c0 = np.float32(1.1)
    L = O.Loop(O.OP_SAXPY, O.F32, n, Y, X=X, c0=c0)
    out = O.run_seq(L)[1]
    two = [rn32(F(rn32(F(c0) * F(x))) + F(y)) for x, y in zip(X, Y)]
    fused = [rn32(F(c0) * F(x) + F(y)) for x, y in zip(X, Y)]
    assert out.tobytes() == np.array(two, dtype=np.float32).tobytes()
    assert sum(a != b for a, b in zip(two, fused)) > 0  # the pin discriminates FMA
    # numpy's float32 ops (a library routine) agree as well
    assert out.tobytes() == (c0 * X + Y).astype(np.float32).tobytes()


def test_fp32_priv_tmp_closed_form():
    """Y[i] = fl(fl(c0 X[i]) + c1); T'[k] = fl(c0 X[max{i: s[i]=k}]) or T[k]."""
    rng = np.random.default_rng(3)
    n, S = 3000, 64
    X = ((rng.integers(0, 2**23, size=n) * 2.0**-22) - 1).astype(np.float32)
    s = rng.integers(0, S - 3, size=n).astype(np.int32)  # slots S-3..S-1 never written
    T0 = np.arange(S, dtype=np.float32)
    c0, c1 = np.float32(1.1), np.float32(0.3)
    L = O.Loop(O.OP_PRIV_TMP, O.F32, n, np.zeros(n, np.float32), s=s, X=X, T=T0, c0=c0, c1=c1)
    st, Y, T = O.run_seq(L)
    assert st == O.OK
    expY = [rn32(F(rn32(F(c0) * F(x))) + F(c1)) for x in X]
    assert Y.tobytes() == np.array(expY, dtype=np.float32).tobytes()
    last = {}
    for i, k in enumerate(s):
        last[int(k)] = i
    expT = [rn32(F(c0) * F(X[last[k]])) if k in last else T0[k] for k in range(S)]
    assert T.tobytes() == np.array(expT, dtype=np.float32).tobytes()
    # profile: no RAW, WAR = WAW = n - |distinct(s)|
    p = O.profile(L)
    d = len(set(s.tolist()))
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (0, n - d, n - d)
    # privatized semantics == sequential (d_raw = 0)
    st, Y2, T2 = O.sim_priv(L)
    assert Y2.tobytes() == Y.tobytes() and T2.tobytes() == T.tobytes()


def test_doall_order_independence():
    """If all three densities are 0, any execution order gives the forward result."""
    rng = np.random.default_rng(11)
    n = 500
    pi = rng.permutation(n).astype(np.int32)
    L = O.Loop(O.OP_ADD_C, O.F32, n, rng.standard_normal(n).astype(np.float32), r=pi, w=pi, c0=np.float32(0.7))
    p = O.profile(L)
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (0, 0, 0)
    fwd = O.run_seq(L)[1]
    assert O.run_order(L, np.arange(n)[::-1].copy())[1].tobytes() == fwd.tobytes()
    assert O.run_order(L, rng.permutation(n))[1].tobytes() == fwd.tobytes()


def test_index_error_no_side_effects():
    A0 = np.arange(8, dtype=np.int32)
    L = O.Loop(O.OP_ADD_C, O.I32, 8, A0, r=np.array([0, 1, 2, 3, 4, 5, 6, 8], np.int32), w=np.arange(8), c0=1)
    st, A, _ = O.run_seq(L)
    assert st == O.ERR_INDEX and A.tolist() == A0.tolist()
    assert O.profile(L)["status"] == O.ERR_INDEX
    L = O.Loop(O.OP_ADD_C, O.I32, 8, A0, r=np.arange(8), w=np.array([0, 1, 2, 3, 4, 5, 6, -1], np.int32), c0=1)
    assert O.sim_tls(L, 4)[0] == O.ERR_INDEX
    # identity index with n > len is out of range too
    L = O.Loop(O.OP_ADD_C, O.I32, 9, A0, c0=1)
    assert O.run_seq(L)[0] == O.ERR_INDEX


def test_window_policy_values():
    """Reading A8: values worked by hand."""
    n = 1 << 24
    assert O.tls_next_window(n, -1, -1) == 4096          # no profile
    assert O.tls_next_window(n, 0, -1) == 65536          # profile says DOALL-like
    assert O.tls_next_window(n, n // 1000, -1) == 4096   # 4n/raw = 4000.2 -> 4096
    assert O.tls_next_window(n, n // 10, -1) == 64       # 40.0 -> 64
    assert O.tls_next_window(n, n, -1) == 32             # 4 -> clamp 32
    assert O.tls_next_window(n, 5, 7, 65536) == 32       # 2*max(7,16) = 32
    assert O.tls_next_window(n, 5, 100, 65536) == 256
    assert O.tls_next_window(n, 5, 4096, 65536) == 8192  # clean window doubles
    assert O.tls_next_window(n, 5, 65536, 65536) == 65536
    assert O.tls_next_window(n, 5, 3000, 1024) == 1024   # cap


def test_adaptive_tls_equals_sequential():
    rng = np.random.default_rng(5)
    n = 3000
    r = rng.integers(0, n, size=n).astype(np.int32)
    w = rng.permutation(n).astype(np.int32)
    L = O.Loop(O.OP_ADD_C, O.I32, n, rng.integers(0, 100, n), r=r, w=w, c0=3)
    seq = O.run_seq(L)[1]
    raw = O.profile(L)["raw_iters"]
    for prof in (-1, raw):
        st, A, _, stats = O.sim_tls(L, 0, 256, prof)
        assert A.tolist() == seq.tolist() and stats["committed"] == n


# ----------------------------------------------------------------------------
# TLS with on-chip recovery (reading B7): jpo_sim_tls_fwd
# ----------------------------------------------------------------------------
def _sub_loop(L, b, e):
    """Iterations [b, e) of L as a loop of their own (index arrays sliced)."""
    sl = lambda a: None if a is None else a[b:e]  # noqa: E731
    return O.Loop(L.op, L.dtype, e - b, L.A, r=sl(L.r), r2=sl(L.r2), w=sl(L.w), s=sl(L.s), X=L.X, T=L.T,
                  c0=L.c0, c1=L.c1)


def test_tls_fwd_golden(golden_dir):
    rows = {g["name"]: g for g in load_golden(golden_dir)}
    with open(os.path.join(golden_dir, "tls_fwd_n8.txt")) as f:
        for line in f:
            if line.startswith("#") or not line.strip():
                continue
            name, nums = [t.strip() for t in line.split("|")]
            W, windows, viol, executed, committed = (int(t) for t in nums.split())
            g = rows[name]
            L = O.Loop(g["op"], O.I32, 8, g["A0"], r=g["r"], r2=g["r2"], w=g["w"], c0=g["c0"])
            st, A, _, stats = O.sim_tls_fwd(L, W)
            assert st == O.OK
            assert A.tolist() == g["A"].tolist(), name
            assert (stats["windows"], stats["violations"], stats["executed"], stats["committed"]) == \
                (windows, viol, executed, committed), name


def test_tls_fwd_exhaustive():
    """N=5, |A|=3, every (r, w), W in {1,2,3,5}: arrays == sequential; the
    violations of each window are the raw iterations of that window taken as a
    loop of its own (jpo_profile_run: a different algorithm); W=1 never
    violates; W >= n gives the whole loop's raw_iters."""
    n, la = 5, 3
    A0 = np.array([5, -3, 11], dtype=np.int32)
    for rw in itertools.product(range(la), repeat=2 * n):
        L = O.Loop(O.OP_ADD_C, O.I32, n, A0, r=np.array(rw[:n], np.int32), w=np.array(rw[n:], np.int32), c0=7)
        seq = O.run_seq(L)[1]
        for W in (1, 2, 3, 5):
            st, A, _, s = O.sim_tls_fwd(L, W)
            assert st == O.OK and A.tolist() == seq.tolist()
            viol = sum(O.profile(_sub_loop(L, b, min(b + W, n)))["raw_iters"] for b in range(0, n, W))
            assert s == {"committed": n, "executed": n + viol, "windows": -(-n // W), "violations": viol}
            if W == 1:
                assert viol == 0
            if W >= n:
                assert viol == O.profile(L)["raw_iters"]


@pytest.mark.parametrize("op", [O.OP_ADD_C, O.OP_STENCIL2, O.OP_SAXPY, O.OP_PRIV_TMP])
@pytest.mark.parametrize("dtype", [O.I32, O.F32])
def test_tls_fwd_random_vs_bruteforce(op, dtype):
    """Random small loops of every opcode: arrays == sequential, and the
    violation count equals the pure-Python pair brute force restricted to
    in-window pairs (j < i in the same window, W(j) ∩ R_exp(i) != {})."""
    rng = np.random.default_rng(100 + op * 2 + dtype)
    for trial in range(20):
        n = int(rng.integers(1, 60))
        la = int(rng.integers(1, 12))
        W = int(rng.integers(1, 20))
        r, r2, w = (rng.integers(0, la, n).astype(np.int32) for _ in range(3))
        s = rng.integers(0, 4, n).astype(np.int32)
        el = np.int32 if dtype == O.I32 else np.float32
        A0 = (rng.integers(-50, 50, la) if dtype == O.I32 else rng.uniform(-1, 1, la)).astype(el)
        X = (rng.integers(-50, 50, la) if dtype == O.I32 else rng.uniform(-1, 1, la)).astype(el)
        T0 = np.zeros(4, dtype=el)
        kw = dict(r=r, w=w)
        if op == O.OP_STENCIL2:
            kw["r2"] = r2
        if op in (O.OP_SAXPY, O.OP_PRIV_TMP):
            kw["X"] = X
        if op == O.OP_PRIV_TMP:
            kw.update(s=s, T=T0)
        c0 = 3 if dtype == O.I32 else np.float32(1.1)
        L = O.Loop(op, dtype, n, A0, c0=c0, c1=(2 if dtype == O.I32 else np.float32(0.3)), **kw)
        _, Aseq, Tseq = O.run_seq(L)
        st, A, T, stats = O.sim_tls_fwd(L, W)
        assert st == O.OK
        assert A.tobytes() == Aseq.tobytes()
        if op == O.OP_PRIV_TMP:
            assert T.tobytes() == Tseq.tobytes()
        sets = [acc_sets(op, i, r, kw.get("r2"), w, kw.get("s")) for i in range(n)]
        viol = sum(any(set(sets[j][2]) & set(sets[i][0]) for j in range((i // W) * W, i)) for i in range(n))
        assert stats == {"committed": n, "executed": n + viol, "windows": -(-n // W), "violations": viol}


def test_tls_fwd_density_zero_and_args():
    """d_raw = 0 (a permutation self-update) => no violations at any W; W = 0 is rejected."""
    n = 300
    perm = np.random.default_rng(5).permutation(n).astype(np.int32)
    L = O.Loop(O.OP_ADD_C, O.I32, n, np.arange(n), r=perm, w=perm, c0=1)
    for W in (1, 7, 64, 1000):
        assert O.sim_tls_fwd(L, W)[3]["violations"] == 0
    assert O.sim_tls_fwd(L, 0)[0] == -1

"""Path 9 (reading B14): one-window on-chip TLS over ADD_C loops WITH WAR / WAW,
the violators fed from the last earlier writer of their address (the profile's
last-writer pass), last writers committing at once or after the window's one
barrier.  Every byte of A against jpo_run_seq and the statistics against
jpo_sim_tls_fwd with W = n (one window, violations = raw iterations).

Expected values come only from oracle/ on the same seeded inputs.
"""
import numpy as np
import pytest
import torch

import oracle as O
import synth
from helpers import random_loop, to_oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = None
    DEV = None


def equal_bytes(t: torch.Tensor, a: np.ndarray) -> bool:
    return torch.equal(t.cpu().view(torch.int32), torch.from_numpy(a.view(np.int32)))


def first_diff(t: torch.Tensor, a: np.ndarray):
    return np.flatnonzero(t.cpu().numpy().view(np.int32) != a.view(np.int32))[:10]


def run_and_check(wl, expect_path=9, **kw):
    ref = to_oracle(wl)
    _, A, _ = O.run_seq(ref)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), **kw)
    torch.cuda.synchronize()
    assert equal_bytes(g.A, A), (first_diff(g.A, A), res)
    if expect_path is not None:
        assert res["mode"] == jp.JP_MODE_TLS and res["tls_path"] == expect_path, res
    if res["tls_path"] == 9:
        assert res["tls_recovery"] == jp.JP_TLS_ONCHIP and res["tls"]["windows"] == 1
        _, A2, _, stats = O.sim_tls_fwd(ref, max(wl.n, 1))
        assert res["tls"] == stats, (res["tls"], stats)
        assert equal_bytes(g.A, A2)
    return res


@pytest.mark.parametrize("d,delta", [(0.001, 1024), (0.01, 1024), (0.05, 1024), (0.10, 1024),
                                     (0.01, 1 << 20), (0.10, 1 << 20)])
def test_config3_waw_full_size_one_window(d, delta):
    """Config 3's shape with WAW at N = 2^24 (the bench's config3_waw rows)."""
    wl = synth.config3_waw(d, delta=delta)
    res = run_and_check(wl)
    p = O.profile(to_oracle(wl))
    assert (res["prof"]["raw_iters"], res["prof"]["waw_iters"]) == (p["raw_iters"], p["waw_iters"])


@pytest.mark.parametrize("seed", [1, 2, 3])
@pytest.mark.parametrize("dtype", [0, 1], ids=["i32", "f32"])
def test_random_raw_war_waw(seed, dtype):
    """Random r and w over len_A = n (RAW, WAR and WAW all present, d_raw ~ 0.37),
    ragged n: exposed reads of later-written addresses exercise the commits after
    the barrier."""
    n = (1 << 20) + 77 * seed
    wl = random_loop(100 + seed, O.OP_ADD_C, dtype, n, len_a=n, null_prob=0.0)
    res = run_and_check(wl)
    assert res["prof"]["war_iters"] > 0 and res["prof"]["waw_iters"] > 0


@pytest.mark.parametrize("frac", [0.5, 0.9])
def test_inplace_mix(frac):
    """In-place updates (r[i] == w[i]: one access record for read and write in the
    profile) mixed with random reads and duplicate writes: path 9 reads the
    also-read records as reads."""
    n = (1 << 20) + 11
    g = np.random.default_rng(17)
    w = g.integers(0, n, n).astype(np.int32)
    r = np.where(g.random(n) < frac, w, g.integers(0, n, n)).astype(np.int32)
    A = torch.from_numpy(g.integers(-2**31, 2**31, size=n, dtype=np.int64).astype(np.int32))
    wl = synth.Workload("inplace_mix", O.OP_ADD_C, O.I32, n, A, r=torch.from_numpy(r), w=torch.from_numpy(w), c0=5)
    res = run_and_check(wl)
    assert res["prof"]["waw_iters"] > 0, res["prof"]


@pytest.mark.parametrize("dtype", [0, 1], ids=["i32", "f32"])
@pytest.mark.parametrize("dup", [0.3, 0.7, 0.9])
def test_saxpy_scatter_add(dtype, dup):
    """SAXPY with duplicate indirect writes, Y[w[i]] = c0*X[r[i]] + Y[w[i]] (a
    scatter-add: the writers of one address form a dependence chain, raw = waw):
    path 9 feeds every later writer from its address's previous writer.  At
    dup = 0.7 a bucket of 8192 addresses gets ~27K writes (the one-CTA-per-SM
    tier of the last-writer pass); at 0.9 ~82K, more than that tier holds: the
    windowed paths run instead (same bytes)."""
    n = (1 << 20) + 29
    g = np.random.default_rng(23 + int(10 * dup))
    m = int(n * (1 - dup)) + 1       # fewer distinct targets -> more duplicates
    w = g.integers(0, m, n).astype(np.int32)
    r = g.integers(0, n, n).astype(np.int32)
    if dtype == O.I32:
        Y = torch.from_numpy(g.integers(-2**31, 2**31, size=n, dtype=np.int64).astype(np.int32))
        X = torch.from_numpy(g.integers(-2**31, 2**31, size=n, dtype=np.int64).astype(np.int32))
        c0 = 3
    else:
        Y = torch.from_numpy(((g.integers(0, 2**23, size=n) * 2.0**-22) - 1).astype(np.float32))
        X = torch.from_numpy(((g.integers(0, 2**23, size=n) * 2.0**-22) - 1).astype(np.float32))
        c0 = float(np.float32(1.1))
    wl = synth.Workload("scatter_add", O.OP_SAXPY, dtype, n, Y, r=torch.from_numpy(r), w=torch.from_numpy(w),
                        X=X, c0=c0)
    res = run_and_check(wl, expect_path=9 if dup < 0.8 else None)
    assert res["prof"]["raw_iters"] == res["prof"]["waw_iters"] > 0, res["prof"]
    if dup > 0.8:
        assert res["tls_path"] != 9, res


def _war_only(n: int, k: int, seed: int = 5):
    """w[i] = r[i-1] (every write lands on an address an EARLIER iteration read,
    no earlier writer: WAR on the window-start value, no WAW), and k iterations
    read what an earlier iteration wrote (RAW, so Fig. 2(b) gives TLS)."""
    g = np.random.default_rng(seed)
    pi = g.permutation(n).astype(np.int32)
    r = pi.copy()
    w = np.roll(pi, 1)
    w[0] = pi[-1]
    dep = np.sort(g.choice(np.arange(4, n), size=k, replace=False))
    r[dep] = w[dep - 3]
    A = torch.from_numpy(g.integers(-2**31, 2**31, size=n, dtype=np.int64).astype(np.int32))
    return synth.Workload("war_only", O.OP_ADD_C, O.I32, n, A, r=torch.from_numpy(r), w=torch.from_numpy(w), c0=7)


def test_war_only_commits_after_barrier():
    n = (1 << 20) + 5
    wl = _war_only(n, 3000)
    res = run_and_check(wl)
    assert res["prof"]["waw_iters"] == 0 and res["prof"]["war_iters"] > n // 2, res["prof"]


def test_hot_address_falls_back():
    """An address written by more writers than the last-writer pass holds (a
    running-sum slot): the windowed restart path runs instead; same bytes."""
    n = 1 << 20
    g = np.random.default_rng(11)
    r = g.integers(0, n, size=n).astype(np.int32)
    w = g.permutation(n).astype(np.int32)
    hot = g.choice(n, size=6000, replace=False)
    w[hot] = 17
    r[hot[::7]] = 17
    A = torch.from_numpy(g.integers(-2**31, 2**31, size=n, dtype=np.int64).astype(np.int32))
    wl = synth.Workload("hot", O.OP_ADD_C, O.I32, n, A, r=torch.from_numpy(r), w=torch.from_numpy(w), c0=3)
    res = run_and_check(wl, expect_path=None)
    assert res["tls_path"] != 9, res


def test_forced_restart_unchanged():
    """tls_recovery = 1 still runs the restart form (A6) on the same WAW loop."""
    wl = synth.config3_waw(0.01, n=1 << 21, delta=1024)
    res = run_and_check(wl, expect_path=None, tls_recovery=1)
    assert res["tls_recovery"] == jp.JP_TLS_RESTART, res


def test_repeat_same_workspace():
    """Two calls on one workspace (the shadow slots of the first are cleared for
    the second), and a write-once loop after a WAW loop on the same sizes."""
    n = 1 << 20
    wl = synth.config3_waw(0.05, n=n, delta=1024)
    ref = to_oracle(wl)
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    ws = jp.workspace(L)
    exp = ref
    for _ in range(2):
        _, Aexp, _ = O.run_seq(exp)
        res = jp.jp_schedule(L, ws)
        torch.cuda.synchronize()
        assert res["tls_path"] == 9 and equal_bytes(g.A, Aexp), res
        exp = O.Loop(ref.op, ref.dtype, ref.n, Aexp.copy(), r=ref.r, w=ref.w, c0=ref.c0)
    w1 = synth.config3(0.05, n=n)
    _, A1, _ = O.run_seq(to_oracle(w1))
    g1 = w1.to(DEV)
    L1 = jp.Loop.from_workload(g1)
    res = jp.jp_schedule(L1, ws)
    torch.cuda.synchronize()
    assert res["tls_path"] == 8 and equal_bytes(g1.A, A1), res


@pytest.mark.parametrize("split", [2, 3])
def test_ranges_of_config3_waw(split):
    """config3_waw run as consecutive ranges (iter_base = ident_off = the range
    start), each through jp_schedule on the shared arrays: every range is a loop of
    its own (path 9 when it still has raw reads inside it, reads of earlier ranges'
    writes see A); the final A is the sequential one."""
    n = (1 << 21) + 10
    wl = synth.config3_waw(0.05, n=n, delta=1024)
    _, A, _ = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    full = jp.Loop.from_workload(g)
    cuts = [n * k // split for k in range(split + 1)]
    paths = []
    for b, e in zip(cuts[:-1], cuts[1:]):
        part = full.range(b, e)
        res = jp.jp_schedule(part, jp.workspace(part))
        torch.cuda.synchronize()
        paths.append(res["tls_path"])
    assert equal_bytes(g.A, A), first_diff(g.A, A)
    assert 9 in paths, paths


@pytest.mark.parametrize("la_log", [23, 25])
def test_large_A_profile_choice(la_log):
    """A random ADD_C loop over a larger A (2^23: the address-bucket profile;
    2^25: more buckets than the scatter's shared memory holds -> the stamp /
    classify profile): same bytes as the oracle either way, and path 9 / the
    windowed paths as the profile allows."""
    n = 1 << 20
    la = 1 << la_log
    g = np.random.default_rng(31)
    w = g.integers(0, la, n).astype(np.int32)
    r = np.where(g.random(n) < 0.3, np.roll(w, 7), g.integers(0, la, n)).astype(np.int32)
    A = torch.from_numpy(g.integers(-2**31, 2**31, size=la, dtype=np.int64).astype(np.int32))
    wl = synth.Workload("largeA", O.OP_ADD_C, O.I32, n, A, r=torch.from_numpy(r), w=torch.from_numpy(w), c0=9)
    res = run_and_check(wl, expect_path=None)
    assert res["mode"] == jp.JP_MODE_TLS, res


def test_graph_cache_alternating_loops():
    """The profile (and path 9) replay CUDA graphs cached per argument set:
    alternating two loops of the same shape on one workspace, and the same loop
    after its index arrays changed in place (same pointers, new values), must
    give the oracle's bytes every time."""
    n = 1 << 20
    a = synth.config3_waw(0.02, n=n, delta=1024)
    b = synth.config3(0.02, n=n)
    ga, gb = a.to(DEV), b.to(DEV)
    La, Lb = jp.Loop.from_workload(ga), jp.Loop.from_workload(gb)
    ws = jp.workspace(La)
    ea, eb = to_oracle(a), to_oracle(b)
    for rep in range(3):
        for g, L, ref, path in ((ga, La, ea, 9), (gb, Lb, eb, 8)):
            _, A, _ = O.run_seq(ref)
            res = jp.jp_schedule(L, ws)
            torch.cuda.synchronize()
            assert res["tls_path"] == path and equal_bytes(g.A, A), (rep, res)
            ref.A[:] = A
    # new index values behind the same pointers (the graph replays the new data)
    c = synth.config3_waw(0.05, n=n, delta=64)
    ga.r.copy_(c.r.to(DEV))
    ga.w.copy_(c.w.to(DEV))
    ref = O.Loop(ea.op, ea.dtype, n, ga.A.cpu().numpy().copy(), r=c.r.numpy(), w=c.w.numpy(), c0=ea.c0)
    _, A, _ = O.run_seq(ref)
    res = jp.jp_schedule(La, ws)
    torch.cuda.synchronize()
    assert equal_bytes(ga.A, A), res


@pytest.mark.parametrize("n", [1, 5, 1000, 16384, 16385, 40000])
@pytest.mark.parametrize("kind", ["write_once", "waw"])
def test_small_n_large_A(n, kind):
    """Few iterations over a large A (the address-bucket profile with one or two
    tiles, a partial last quad, most buckets empty): same bytes as the oracle."""
    la = 1 << 20
    g = np.random.default_rng(n + (7 if kind == "waw" else 0))
    if kind == "write_once":
        w = g.choice(la, size=n, replace=False).astype(np.int32)
    else:
        w = g.integers(0, max(2, n // 2), n).astype(np.int32)
    r = w.copy()
    dep = g.random(n) < 0.2
    src = np.maximum(np.arange(n) - 1 - g.integers(0, 50, n), 0)
    r[dep] = w[src[dep]]
    r[0] = w[0]
    A = torch.from_numpy(g.integers(-2**31, 2**31, size=la, dtype=np.int64).astype(np.int32))
    wl = synth.Workload("small_n", O.OP_ADD_C, O.I32, n, A, r=torch.from_numpy(r), w=torch.from_numpy(w), c0=11)
    run_and_check(wl, expect_path=None)

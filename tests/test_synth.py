"""Generator tests: counter-based draws, determinism, and designed densities."""
import numpy as np
import pytest
import torch

import oracle as O
import synth
from synth.gen import rnd, splitmix64

M = (1 << 64) - 1


def sm_ref(x):
    x = (x + 0x9E3779B97F4A7C15) & M
    x = ((x ^ (x >> 30)) * 0xBF58476D1CE4E5B9) & M
    x = ((x ^ (x >> 27)) * 0x94D049BB133111EB) & M
    return x ^ (x >> 31)


def test_splitmix64_matches_python_ints():
    xs = [0, 1, 2, 12345, (1 << 63) - 1, 1 << 63, M, 0xDEADBEEFCAFEBABE]
    t = torch.tensor([x - (1 << 64) if x >= 1 << 63 else x for x in xs], dtype=torch.int64)
    got = [int(v) & M for v in splitmix64(t)]
    assert got == [sm_ref(x) for x in xs]
    # splitmix64 of 0 after one increment is the well-known first output of seed 0
    assert sm_ref(0) == 0xE220A8397B1DCDAF
    r = rnd(1003, 5, torch.arange(4, dtype=torch.int64))
    assert [int(v) & M for v in r] == [sm_ref(((1003 << 40) ^ (5 << 32) ^ i) & M) for i in range(4)]


def test_f32_data_exact_grid():
    x = synth.f32_data(1002, 2, 10000)
    assert x.dtype == torch.float32
    assert float(x.min()) >= -1.0 and float(x.max()) < 1.0
    k = (x.double() + 1.0) * 2**22
    assert torch.equal(k, k.round())


def test_permutation_is_permutation_and_deterministic():
    p = synth.permutation(7, 5000)
    assert torch.equal(torch.sort(p).values, torch.arange(5000))
    assert torch.equal(p, synth.permutation(7, 5000))
    assert not torch.equal(p, synth.permutation(8, 5000))


def _oracle_loop(wl):
    a = lambda t: None if t is None else t.numpy()  # noqa: E731
    return O.Loop(wl.op, wl.dtype, wl.n, a(wl.A), r=a(wl.r), r2=a(wl.r2), w=a(wl.w), s=a(wl.s), X=a(wl.X),
                  T=a(wl.T), c0=wl.c0, c1=wl.c1)


def test_config1_designed_density():
    for d, k in ((0.0, 0), (0.05, 205)):
        wl = synth.config1(d)
        p = O.profile(_oracle_loop(wl))
        assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (k, 0, 0)


def test_config3_designed_density_reduced():
    for d in (0.001, 0.01, 0.05, 0.10):
        wl = synth.config3(d, n=1 << 16)
        p = O.profile(_oracle_loop(wl))
        assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (round(d * (1 << 16)), 0, 0)


def test_config3_full_size_exact():
    wl = synth.config3(0.01)
    p = O.profile(_oracle_loop(wl))
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (round(0.01 * (1 << 24)), 0, 0)


def test_config4_profile():
    wl = synth.config4(n=1 << 14)
    p = O.profile(_oracle_loop(wl))
    distinct = len(set(wl.s.tolist()))
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (0, (1 << 14) - distinct, (1 << 14) - distinct)


def test_config5_regions():
    n = 1 << 14
    wl = synth.config5(n=n)
    p = O.profile(_oracle_loop(wl))
    assert (p["raw_iters"], p["war_iters"], p["waw_iters"]) == (wl.meta["raw"], wl.meta["war"], wl.meta["waw"])
    f = p["flags"]
    (h0, h1), (m0, m1), (t0, t1) = wl.meta["regions"]
    assert not f[h0:h1].any()                  # head: DOALL
    assert (f[m0:m1] & 6).sum() == 0           # middle: RAW only
    assert (f[t0:t1] & 1).sum() == 0           # tail: no RAW
    assert np.count_nonzero(f[t0:t1] & 4) == n // 8


def test_device_agnostic_bits():
    # the same recipe on the same device twice is bit-identical
    a = synth.config4(n=4096)
    b = synth.config4(n=4096)
    for k in ("s", "X", "T", "A"):
        assert torch.equal(getattr(a, k), getattr(b, k))


@pytest.mark.parametrize("d,delta", [(0.0, 1024), (0.01, 1024), (0.1, 64), (0.05, 1 << 20)])
def test_config3_waw_designed_profile(d, delta):
    """The WAW variant of config 3: raw = K exactly, waw = n/2 exactly (every
    address of [0, n/2) written twice), against the oracle's profile."""
    n = 1 << 13
    wl = synth.config3_waw(d, n=n, delta=delta)
    p = O.profile(_oracle_loop(wl))
    assert (p["raw_iters"], p["waw_iters"]) == (wl.meta["raw"], n // 2)
    assert wl.meta["raw"] == round(d * n)
    assert int(wl.w.max()) < n // 2 and int(wl.r.max()) < n

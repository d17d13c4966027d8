"""The static check's affine sample riding on the address-bucket profile's first
kernel (jp_schedule, A >= 2^20): when the sample looks affine the rest of the
profile exits at once and the full static check decides (reading B8); otherwise
the profile's result stands.  Every case ends in the sequential state (oracle).
"""
import numpy as np
import pytest
import torch

import oracle as O
import synth
from helpers import to_oracle

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = None
    DEV = None

N = (1 << 20) + 37


def _loop(r, w, dtype=O.I32, seed=3):
    g = np.random.default_rng(seed)
    n = len(r)
    la = int(max(r.max(), w.max()) + 1)
    if dtype == O.I32:
        A = torch.from_numpy(g.integers(-2**31, 2**31, size=la, dtype=np.int64).astype(np.int32))
        c0 = 7
    else:
        A = torch.from_numpy(((g.integers(0, 2**23, size=la) * 2.0**-22) - 1).astype(np.float32))
        c0 = float(np.float32(1.1))
    return synth.Workload("affine", O.OP_ADD_C, dtype, n, A, r=torch.from_numpy(r.astype(np.int32)),
                          w=torch.from_numpy(w.astype(np.int32)), c0=c0)


def _run(wl, **kw):
    _, A, _ = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    res = jp.jp_schedule(L, jp.workspace(L), **kw)
    torch.cuda.synchronize()
    assert torch.equal(g.A.cpu().view(torch.int32), torch.from_numpy(A.view(np.int32))), res
    return res


@pytest.mark.parametrize("dtype", [O.I32, O.F32])
def test_affine_independent_is_doall_unprofiled(dtype):
    """r[i] = 2i + 1, w[i] = 2i (disjoint lattices): DOALL with no profile."""
    i = np.arange(N, dtype=np.int64)
    res = _run(_loop(2 * i + 1, 2 * i, dtype))
    assert res["mode"] == jp.JP_MODE_DOALL and res["profiled"] == 0, res


def test_affine_dependent_runs_the_profile():
    """r[i] = i, w[i] = i + 1: affine but every iteration reads its predecessor's
    write (a chain): the sample looks affine, the full check finds the conflict,
    the profile runs and Fig. 2(b) decides."""
    i = np.arange(N, dtype=np.int64)
    res = _run(_loop(i, i + 1))
    assert res["profiled"] == 1 and res["prof"]["raw_iters"] == N - 1, res


def test_affine_prefix_only():
    """Affine on the first 64 entries only: the sample looks affine, the full pass
    says not affine, the profile runs."""
    g = np.random.default_rng(5)
    r = g.permutation(N).astype(np.int64)
    w = r.copy()
    r[:100] = np.arange(100)
    w[:100] = np.arange(100)
    # keep w a permutation: move the displaced values out of the prefix
    res = _run(_loop(r, w))
    assert res["profiled"] == 1, res


def test_random_runs_the_profile_as_before():
    """Config 3 (random indices): the sample fails on the device, the profile that
    was queued behind it stands (path 8), and the result is the oracle's."""
    wl = synth.config3(0.01, n=N)
    res = _run(wl)
    assert res["profiled"] == 1 and res["tls_path"] == 8, res


def test_static_check_off_profiles_affine():
    i = np.arange(N, dtype=np.int64)
    res = _run(_loop(2 * i + 1, 2 * i), static_check=1)
    assert res["profiled"] == 1 and res["mode"] == jp.JP_MODE_DOALL, res

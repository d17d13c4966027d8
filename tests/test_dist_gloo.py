"""Multi-process (gloo, CPU) tests of the multi-GPU driver dist.py.

world_size 2 and 3 processes on 127.0.0.1; every rank holds full-size
replicas and its task-sharing range.  The compute entry points are the test
double in tests/fake_engine.py (numpy over the REAL workspace layout), so these
tests exercise the collectives (C1 MAX int32 tables, C3 SUM counts, C4 MAX int64
packed keys, TLS broadcast) and the plan exactly as on the GPUs, and compare
with the oracle's sequential result.
"""
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _sharing_case(rank, world, case, q, exchange="dense"):
    try:
        import fake_engine as fe
        import oracle as O
        import paper_conf_icpp_hanzlw13_b200 as jp
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth
        from helpers import region_workload, to_oracle

        wl = {"c1_0": lambda: synth.config1(0.0, n=600), "c1_5": lambda: synth.config1(0.05, n=600),
              "c4": lambda: synth.config4(n=700, slots=64), "c3": lambda: synth.config3(0.02, n=512),
              "c2": lambda: synth.config2(n=901), "c5tail": lambda: region_workload(synth.config5(n=1 << 11), 3 << 9, 1 << 11),
              "c5head": lambda: region_workload(synth.config5(n=1 << 11), 0, 1 << 10)}[case]()
        ref = to_oracle(wl)
        _, A_exp, T_exp = O.run_seq(ref)
        p_exp = O.profile(ref)
        full = jp.Loop.from_workload(wl)
        b, e = jd.sharing_ranges(wl.n, world, engine=fe)[rank]
        if case == "c2":   # identity-only: sharded arrays, ident_off = 0
            shard = jp.Loop(wl.op, wl.dtype, e - b, wl.A[b:e].clone(), X=wl.X[b:e].clone(), c0=wl.c0,
                            iter_base=b)
            jd.schedule_partitioned(shard, None, engine=fe)
            ok = shard.tensors["A"].numpy().tobytes() == A_exp[b:e].tobytes()
            q.put((rank, ok, None))
            return
        loop = full.range(b, e)
        ws = torch.zeros(jp.jp_workspace_bytes(loop), dtype=torch.uint8)
        jd.OWNER_MIN_LEN = 0   # small test tables still take the owner form
        res = jd.schedule_partitioned(loop, ws, full_loop=full, engine=fe, exchange=exchange)
        prof_ok = (res["prof"]["raw_iters"], res["prof"]["war_iters"], res["prof"]["waw_iters"],
                   res["prof"]["first_raw_iter"]) == (p_exp["raw_iters"], p_exp["war_iters"], p_exp["waw_iters"],
                                                      p_exp["first_raw_iter"])
        ok_A = wl.A.numpy().tobytes() == A_exp.tobytes()
        if wl.op == O.OP_PRIV_TMP:   # Y identity-indexed: sharded; T keyed: replicated
            ok_A = wl.A.numpy()[b:e].tobytes() == A_exp[b:e].tobytes()
            ok_A &= wl.T.numpy().tobytes() == T_exp.tobytes()
        q.put((rank, bool(prof_ok and ok_A), res["mode_name"]))
    except Exception as ex:  # pragma: no cover - reported to the parent
        q.put((rank, False, repr(ex)))


def _group_worker(rank, world, port, jobs, q):
    """One process group per world size; every job (a test case) runs in it in turn."""
    sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        for k, (kind, case, exchange) in enumerate(jobs):
            sub = _Tagged(q, k)
            if kind == "share":
                _sharing_case(rank, world, case, sub, exchange)
            else:
                _steal_case(rank, world, case, exchange, sub)
            dist.barrier()
    finally:
        dist.destroy_process_group()


class _Tagged:
    def __init__(self, q, k):
        self.q, self.k = q, k

    def put(self, item):
        self.q.put((self.k, item))


_RESULTS = {}


def _jobs(world):
    if world == 4:
        return [("share", "c4", "dense"), ("share", "c4", "owner"), ("share", "c5tail", "owner"),
                ("share", "c3", "owner"), ("steal", "c5", "owner")]
    share = [("share", c, "dense") for c, _ in _CASES]
    if world == 3:
        share += [("share", c, "owner") for c in ("c1_5", "c4", "c5tail", "c5head")]
    else:
        share += [("share", "c5tail", "owner")]
    steal = [("steal", "c5", "dense"), ("steal", "c5", "owner"), ("steal", "c5", "dense+repl")] + \
        ([("steal", "c1_5", "dense"), ("steal", "seq", "dense"), ("steal", "c5", "owner+repl"),
          ("steal", "seq", "dense+repl")] if world == 2 else [])
    return share + steal


def run_world(world, kind, case, exchange="dense"):
    """Results of one case; the whole world-size group runs once and is cached."""
    if world not in _RESULTS:
        jobs = _jobs(world)
        ctx = mp.get_context("spawn")
        q = ctx.Queue()
        port = _free_port()
        ps = [ctx.Process(target=_group_worker, args=(r, world, port, jobs, q)) for r in range(world)]
        for p in ps:
            p.start()
        got = {}
        for _ in range(world * len(jobs)):
            k, item = q.get(timeout=600)
            got.setdefault(jobs[k], []).append(item)
        for p in ps:
            p.join(timeout=60)
        _RESULTS[world] = {j: sorted(v, key=lambda x: x[0]) for j, v in got.items()}
    return _RESULTS[world][(kind, case, exchange)]


_CASES = [("c1_0", "DOALL"), ("c1_5", "TLS"), ("c4", "PRIVATIZED"), ("c3", "TLS"), ("c2", None),
          ("c5tail", "PRIVATIZED"), ("c5head", "DOALL")]


@pytest.mark.parametrize("world,case,mode,exchange",
                         [(w, c, m, "dense") for w in (2, 3) for c, m in _CASES] +
                         [(3, c, m, "owner") for c, m in _CASES if c in ("c1_5", "c4", "c5tail", "c5head")] +
                         [(2, "c5tail", "PRIVATIZED", "owner")] +
                         [(4, "c4", "PRIVATIZED", "dense"), (4, "c4", "PRIVATIZED", "owner"),
                          (4, "c5tail", "PRIVATIZED", "owner"), (4, "c3", "TLS", "owner")])
def test_partitioned_schedule_matches_oracle(world, case, mode, exchange):
    out = run_world(world, "share", case, exchange)
    assert [o[1] for o in out] == [True] * world, out
    if mode:
        assert all(o[2] == mode for o in out), out


def test_sharing_ranges_cover_and_match_plan():
    import fake_engine as fe
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    rg = jd.sharing_ranges(1 << 28, 8, engine=fe)
    assert rg[0][0] == 0 and rg[-1][1] == 1 << 28 and all(e - s == 1 << 25 for s, e in rg)
    chunks, stolen = jd.stealing_plan([(0, 1 << 20, 2), (1 << 20, 1 << 22, 0)], 4, 1 << 16, engine=fe)
    assert all(c[3] == 0 for c in chunks if c[2] == 2)
    assert np.sum([c[1] - c[0] for c in chunks]) == 1 << 22


def _steal_case(rank, world, case, exchange, q):
    try:
        import fake_engine as fe
        import oracle as O
        import paper_conf_icpp_hanzlw13_b200 as jp
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth
        from helpers import to_oracle
        from helpers import seq_mixed
        wl = {"c5": lambda: synth.config5(n=1 << 12, delta=64),
              "c1_5": lambda: synth.config1(0.05, n=4096), "seq": lambda: seq_mixed(3 * 1024)}[case]()
        ref = to_oracle(wl)
        _, A_exp, _ = O.run_seq(ref)
        full = jp.Loop.from_workload(wl)
        ws = torch.zeros(jp.jp_workspace_bytes(full), dtype=torch.uint8)
        jd.OWNER_MIN_LEN = 0
        # "<exchange>+repl": every rank profiles its full replica (jp_profile_plan_tasks);
        # otherwise the partitioned profile with C1 / C3
        xch, _, repl = exchange.partition("+")
        res = jd.schedule_stealing(full, ws, chunk_iters=1024, exchange=xch, engine=fe,
                                   profile="replicated" if repl else "partitioned")
        ok = wl.A.numpy().tobytes() == A_exp.tobytes()
        q.put((rank, bool(ok), res["n_tasks"], res["n_batches"], res["rank_work"]["iters"]))
    except Exception:  # pragma: no cover
        import traceback
        q.put((rank, False, traceback.format_exc(), 0, 0))


@pytest.mark.parametrize("case,world,exchange", [("c5", 2, "dense"), ("c5", 3, "dense"), ("c5", 2, "owner"),
                                                  ("c5", 3, "owner"), ("c1_5", 2, "dense"), ("seq", 2, "dense"),
                                                  ("c5", 4, "owner"), ("c5", 2, "dense+repl"),
                                                  ("c5", 3, "dense+repl"), ("c5", 2, "owner+repl"),
                                                  ("seq", 2, "dense+repl")])
def test_stealing_scheme_matches_oracle(case, world, exchange):
    """Multi-rank task stealing (dist.schedule_stealing): partitioned profile with
    chunk counts (or, "+repl", every rank's own profile of its full replica),
    tasks + PDG, Alg. 1 plan, batches with C4 merges; every replica ends with the
    oracle's sequential result."""
    out = run_world(world, "steal", case, exchange)
    assert [o[1] for o in out] == [True] * world, out
    assert sum(o[4] for o in out) == (3 * 1024 if case == "seq" else 4096)

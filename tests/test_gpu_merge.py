"""C4 fused into the privatized stream (jp_priv_stream_merge, dist.PrivMerge):
config 4's rank ranges streamed, the 1024 last-writer keys pushed into every
rank's inbox over peer memory and merged + applied inside the same kernel.
Compared with the oracle (jpo_run_seq) byte for byte: T on every rank, Y on the
range each rank ran; over several epochs (the parity double buffer) and through
a CUDA-graph replay."""
import multiprocessing as mp
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist

import oracle as O
import synth
from helpers import to_oracle

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

if torch.cuda.is_available():
    import paper_conf_icpp_hanzlw13_b200 as jp
    from paper_conf_icpp_hanzlw13_b200 import dist as jd
    DEV = torch.device("cuda:0")
else:  # collected on CPU boxes, never run there
    jp = jd = None
    DEV = None


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.mark.parametrize("n,slots", [((1 << 20) + 77, 1024), (4096 * 3 + 5, 32), (5000, 4096)])
def test_fused_merge_one_rank(n, slots):
    wl = synth.config4(n=n, slots=slots)
    _, A_exp, T_exp = O.run_seq(to_oracle(wl))
    g = wl.to(DEV)
    T0, A0 = g.T.clone(), g.A.clone()
    full = jp.Loop.from_workload(g)
    loop = full.range(0, n)
    ws = jp.workspace(loop)
    m = jd.PrivMerge(loop, ws)
    for _ in range(3):   # epochs 1..3 (both parities)
        g.T.copy_(T0)
        g.A.copy_(A0)
        m.step()
        m.check()
        assert g.T.cpu().numpy().tobytes() == T_exp.tobytes()
        assert g.A.cpu().numpy().tobytes() == A_exp.tobytes()
    gr = m.graph()
    if gr is not None:   # the same step replayed from a CUDA graph
        for _ in range(2):
            g.T.copy_(T0)
            g.A.copy_(A0)
            gr.replay()
            m.check()
            assert g.T.cpu().numpy().tobytes() == T_exp.tobytes()
            assert g.A.cpu().numpy().tobytes() == A_exp.tobytes()
    m.close()


def test_fused_merge_rejects_other_shapes():
    wl = synth.config4(n=1 << 14)
    wl.w = torch.arange(wl.n, dtype=torch.int32)   # Y through an index: not the fused shape
    g = wl.to(DEV)
    L = jp.Loop.from_workload(g)
    assert jp.jp_priv_inbox_bytes(L, 1) == 0
    with pytest.raises(ValueError):
        jd.PrivMerge(L, jp.workspace(L))


def _worker(rank, world, port, q):
    sys.path[:0] = [ROOT, os.path.join(ROOT, "tests")]
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle as O
        import paper_conf_icpp_hanzlw13_b200 as jp
        from paper_conf_icpp_hanzlw13_b200 import dist as jd
        import synth
        from helpers import to_oracle
        wl = synth.config4(n=(1 << 18) + 64, slots=1024)
        _, A_exp, T_exp = O.run_seq(to_oracle(wl))
        g = wl.to("cuda:0")
        T0, A0 = g.T.clone(), g.A.clone()
        full = jp.Loop.from_workload(g)
        b, e = jd.sharing_ranges(wl.n, world)[rank]
        loop = full.range(b, e)
        ws = jp.workspace(loop)
        m = jd.PrivMerge(loop, ws)
        ok = True
        for _ in range(3):
            g.T.copy_(T0)
            g.A.copy_(A0)
            torch.cuda.synchronize()
            dist.barrier()
            m.step()
            m.check()
            ok &= g.T.cpu().numpy().tobytes() == T_exp.tobytes()
            ok &= g.A.cpu().numpy()[b:e].tobytes() == A_exp[b:e].tobytes()
        dist.barrier()
        m.close()
        q.put((rank, bool(ok)))
    except Exception:  # pragma: no cover
        import traceback
        q.put((rank, traceback.format_exc()))
    finally:
        dist.destroy_process_group()


def test_fused_merge_two_processes():
    """Two ranks (processes) sharing the GPU, inboxes mapped through CUDA IPC."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    ps = [ctx.Process(target=_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in ps:
        p.start()
    out = sorted(q.get(timeout=300) for _ in range(2))
    for p in ps:
        p.join(timeout=120)
    assert out == [(0, True), (1, True)], out

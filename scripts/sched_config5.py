"""Warm jp_schedule(STEALING) calls on config 5 (N = 2^24), for ncu launch lists and timing."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

reps = int(sys.argv[1]) if len(sys.argv) > 1 else 3
wl = synth.config5(device="cuda")
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
for _ in range(reps):
    wl.A.copy_(A0)
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    res = jp.jp_schedule(L, ws, scheme=jp.JP_SCHED_STEALING, chunk_iters=65536)
    torch.cuda.synchronize()
    print(f"{(time.perf_counter() - t0) * 1e3:.3f} ms", res["tls"], res["tls_path"])

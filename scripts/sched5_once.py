#!/usr/bin/env python
"""One config-5 jp_schedule(STEALING) call after a warm-up: for ncu launch lists."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

wl = synth.config5(device="cuda")
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
for _ in range(2):
    wl.A.copy_(A0)
    res = jp.jp_schedule(L, ws, scheme=jp.JP_SCHED_STEALING, chunk_iters=65536)
torch.cuda.synchronize()
print(res["n_tasks"], res["tls_path"], res["tls"])

#!/usr/bin/env python
"""One config3_waw jp_schedule call (d = 1%, path 9) after a warm-up: for ncu launch lists."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

d = float(sys.argv[1]) if len(sys.argv) > 1 else 0.01
wl = synth.config3_waw(d, device="cuda")
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
for _ in range(2):
    wl.A.copy_(A0)
    res = jp.jp_schedule(L, ws)
torch.cuda.synchronize()
print(res["mode_name"], res["tls_path"], res["tls"])

"""One warm jp_schedule() call on config 3 (N = 2^24) at density d, for ncu launch lists.
Usage: python scripts/sched_config3.py [d] [reps]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

d = float(sys.argv[1]) if len(sys.argv) > 1 else 0.01
reps = int(sys.argv[2]) if len(sys.argv) > 2 else 2
wl = synth.config3(d, device="cuda")
A0 = wl.A.clone()
L = jp.Loop.from_workload(wl)
ws = jp.workspace(L)
for _ in range(reps):
    wl.A.copy_(A0)
    res = jp.jp_schedule(L, ws)
torch.cuda.synchronize()
print(res)

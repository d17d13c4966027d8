#!/usr/bin/env python
"""Config 4 on one rank: the fused stream + merge step (jp_priv_stream_merge,
graph replay) vs the plain privatized run; median of 20 (CUDA events)."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import bench  # noqa: E402
import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
from paper_conf_icpp_hanzlw13_b200 import dist as jd  # noqa: E402
import synth  # noqa: E402

st = torch.cuda.current_stream()
wl = synth.config4(device="cuda")
full = jp.Loop.from_workload(wl)
loop = full.range(0, wl.n)
ws = jp.workspace(loop)
prof = jp.jp_profile_density(loop, ws)
m = jd.PrivMerge(loop, ws)
g = m.graph()
_, ms_f = bench.median_timed(g.replay if g else m.step, None, None, st, 20)
_, ms_d = bench.median_timed(m.step, None, None, st, 20)
_, ms_p = bench.median_timed(lambda: jp.jp_run_privatized(loop, prof, ws, stream=st), None, None, st, 20)
m.check()
print(f"fused (graph) {ms_f * 1e3:.1f} us, fused (launch) {ms_d * 1e3:.1f} us, plain privatized {ms_p * 1e3:.1f} us, "
      f"fixed cost {(ms_f - ms_p) * 1e3:.1f} us, graph {g is not None}")

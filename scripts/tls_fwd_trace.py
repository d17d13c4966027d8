#!/usr/bin/env python
"""Per-phase cycle breakdown of the on-chip TLS grid kernel (trace build:
JP_LIB=paper_conf_icpp_hanzlw13_b200/libjp_trace.so).  Marks of CTA 0 / thread 0:
0 start 1 log issued 2 after grid barrier 3 DC resolved 4 non-violators published
5 recovery done 6 commit issued 7 forwarding done 8 next indices issued"""
import ctypes as C
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402

lib = jp.lib()
fn = lib.jp_tls_fwd_trace
fn.argtypes = [C.c_void_p, C.c_int32]
dev = torch.device("cuda:0")
for d in (0.001, 0.1):
    wl = synth.config3(d, device=dev)
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    prof = jp.jp_profile_density(L, ws)
    jp.jp_tls_guide(L, ws)
    for rep in range(2):
        wl.A.copy_(A0)
        torch.cuda.synchronize()
        s = jp.jp_run_tls(L, prof=prof, ws=ws, guided=True, recovery=1, path=6)
        torch.cuda.synchronize()
    buf = np.zeros(2048 * 16, dtype=np.int64)
    fn(buf.ctypes.data, buf.size)
    full = buf.reshape(2048, 16)[2:s["windows"] - 1]
    t = full[:, :9]
    extra = {"first_any_sync": round(float((full[:, 9] - full[:, 4]).mean())), "passes": full[:, 10].tolist()[:20],
             "warp0_pending": full[:, 11].tolist()[:20]}
    dif = np.diff(t, axis=1).mean(axis=0)
    tot = (t[1:, 0] - t[:-1, 0]).mean()
    print(json.dumps({"d": d, "windows": s["windows"], "cycles_per_window": round(float(tot)),
                      "phases": [round(float(x)) for x in dif],
                      "names": ["log", "barrier", "probes+DC", "publish", "recovery", "commit", "forward", "idx"],
                      **extra}))

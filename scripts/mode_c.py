"""Mode C (d_raw > tau_high) on the device: one-warp program-order path (7) vs
TLS with restart (A6) and with on-chip recovery (B7), whole jp_schedule call,
CUDA events.  Usage: python scripts/mode_c.py"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402


def chain(n, gs=False, stride=1):
    ar = torch.arange(n, dtype=torch.int32, device="cuda")
    A = torch.from_numpy(np.random.default_rng(n).integers(0, 1 << 20, size=n).astype(np.int32)).cuda()
    r = torch.clamp(ar - stride, min=0)
    if gs:
        return synth.Workload("gs", 3, 0, n, A, r=r, r2=torch.clamp(ar + 1, max=n - 1), w=ar.clone(), c0=3)
    return synth.Workload("chain", 0, 0, n, A, r=r, w=ar.clone(), c0=7)


def run(wl, **kw):
    A0 = wl.A.clone()
    L = jp.Loop.from_workload(wl)
    ws = jp.workspace(L)
    best, res = None, None
    for _ in range(3):
        wl.A.copy_(A0)
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        res = jp.jp_schedule(L, ws, **kw)
        b.record()
        torch.cuda.synchronize()
        t = a.elapsed_time(b)
        best = t if best is None else min(best, t)
    return {"ms": round(best, 3), "iters_per_s": wl.n / (best * 1e-3), "mode": res["mode_name"],
            "path": res["tls_path"], "windows": res["tls"]["windows"]}


out = {}
for name, mk in (("chain_d100", lambda n: chain(n)), ("gauss_seidel", lambda n: chain(n, gs=True)),
                 ("chain_stride16", lambda n: chain(n, stride=16))):
    row = {"serial_2^20": run(mk(1 << 20)), "restart_2^20": run(mk(1 << 20), tls_recovery=1),
           "serial_2^16": run(mk(1 << 16)), "onchip_2^16": run(mk(1 << 16), tls_recovery=2)}
    out[name] = row
    print(name, row, flush=True)

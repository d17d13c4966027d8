#!/usr/bin/env python
"""Per-phase cycle breakdown of the cluster TLS kernel (trace builds of libjp:
JP_LIB=.../libjp_trace*.so).  Prints mean SM cycles between the phase marks of
CTA 0 / thread 0 over windows 16..2047:
  0 start  1 SE issued  2 after B1  3 DC loads+warp min  4 after B2  5 commit issued
  6 ring wait  7 after B3"""
import json
import os
import sys
import ctypes as C

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_icpp_hanzlw13_b200 as jp  # noqa: E402
import synth  # noqa: E402


def main():
    lib = jp.lib()
    fn = lib.jp_tls_trace
    fn.argtypes = [C.c_void_p, C.c_int32]
    dev = torch.device("cuda:0")
    tag = os.path.basename(os.environ.get("JP_LIB", "libjp.so"))
    for d in [float(x) for x in os.environ.get("TRACE_DENS", "0.001,0.01,0.1").split(",")]:
        wl = synth.config3(d, n=1 << 24, device=dev)
        A0 = wl.A.clone()
        L = jp.Loop.from_workload(wl)
        ws = jp.workspace(L)
        prof = jp.jp_profile_density(L, ws)
        jp.jp_tls_guide(L, ws)
        for path, cl, window, wmax, guided in ((3, 16, 4096, 4096, False), (3, 8, 0, 4096, False),
                                               (3, 8, 0, 4096, True), (1, 0, 4096, 4096, False),
                                               (1, 0, 0, 4096, False), (1, 0, 4096, 4096, True),
                                               (1, 0, 0, 4096, True)):
            for rep in range(2):
                wl.A.copy_(A0)
                torch.cuda.synchronize()
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record()
                s = jp.jp_run_tls(L, window=window, w_max=wmax, path=path, cluster=cl, prof=prof, ws=ws,
                                  guided=guided)
                b.record()
                torch.cuda.synchronize()
            n = 2048 * 16
            buf = np.zeros(n, dtype=np.int64)
            fn(buf.ctypes.data, n)
            t16 = buf.reshape(2048, 16)[16:]
            t = t16[:, :8]
            dif = np.diff(t, axis=1).mean(axis=0)
            tot = (t[1:, 0] - t[:-1, 0]).mean()
            fine = {}
            if path == 1:   # fine marks of the CTA kernel: 0 top, 8 fill, 9 ring reads, 10 gathers, 1 inserts,
                            # 11 fv read, 12 values, 13 loop bookkeeping
                rel = lambda a, b: round(float((t16[:, b] - t16[:, a]).mean()), 0)  # noqa: E731
                fine = {"fill": rel(0, 8), "ring": rel(8, 9), "gather_issue": rel(9, 10), "inserts": rel(10, 1),
                        "fv_to_values": rel(11, 12), "b3_to_book": rel(7, 13),
                        "book_to_next": round(float((t16[1:, 0] - t16[:-1, 13]).mean()), 0)}
            print(json.dumps({"lib": tag, "d": d, "path": path, "guided": guided, "cluster": cl, "window": window, "ms": round(a.elapsed_time(b), 2),
                              "us_per_window": round(a.elapsed_time(b) * 1e3 / s["windows"], 3),
                              "cyc_window": round(float(tot), 0),
                              "cyc_phases": [round(float(x), 0) for x in dif],
                              "cyc_b3_to_next": round(float((t[1:, 0] - t[:-1, 7]).mean()), 0), "fine": fine}),
                  flush=True)


if __name__ == "__main__":
    main()

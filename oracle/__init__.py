"""TEST INFRASTRUCTURE ONLY -- the CPU oracle for the Japonica loop-mode hot path.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package.  The product path
(``paper_conf_icpp_hanzlw13_b200``) never imports it, and the two share no code.
"""
from .oracle import (  # noqa: F401
    OP_ADD_C, OP_SAXPY, OP_PRIV_TMP, OP_STENCIL2, I32, F32, OK, ERR_INDEX,
    Loop, run_seq, run_seq_inplace, run_order, profile, pairs, raw_sources, sim_tls, sim_tls_fwd, tls_next_window, sim_priv, build,
)

"""Seeded synthetic input generators shared by tests, bench.py and smoke().

This module holds NONE of the method's arithmetic: it only draws index arrays
and data with a counter-based generator (splitmix64 finalizer), so that the
oracle side and the CUDA side are fed byte-identical inputs.  Recipes are in
DESIGN.md Sec.5 and follow SURVEY.md Sec.8(d) "Common generator" and the
config table, shaped like the paper's workloads (BASELINE.json configs).
"""
from .gen import (  # noqa: F401
    splitmix64, rnd, permutation, i32_data, f32_data, dependent_set,
    config1, config2, config3, config3_waw, config4, config5, Workload, C0_F32, C1_F32, C0_I32,
    workflow_bicg, workflow_2mm, workflow_crypt, f32_specials, F32_SPECIAL_BITS, dep_region,
)

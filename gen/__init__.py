"""Seeded synthetic inputs shared by the oracle tests and the CUDA path.

Holds NONE of the method's arithmetic (no codes, no SpMV/CG): only the TeaLeaf
matrix recipe G-TEA (TeaLeaf ref [19], P:778-781 — the paper
itself gives only the grid size), random vectors and fault
schedules from a counter-based splitmix64.
"""
from .tealeaf import (tealeaf_csr, tealeaf_rhs, const_k_csr, strip_csr, splitmix64, uniform_pm1, chunk_plan, chunk_csr,  # noqa: F401,E501
                      fault_positions)
from .spd import random_spd_csr  # noqa: F401,E402

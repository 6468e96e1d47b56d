"""B200-native ABFT-protected CG (Pawelczak et al., CLUSTER 2017) — see DESIGN.md.

The product is libabft.so (CUDA for sm_100a behind the C ABI in include/abft.h);
`abft` is its ctypes binding.  Import it explicitly:

    from paper_conf_cluster_pawelczakmpm17_b200 import abft
"""
__all__ = ["abft", "build"]

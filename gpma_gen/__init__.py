"""Seeded synthetic inputs shared by the oracle tests, the CUDA parity tests and bench.py.

This module holds NONE of the method's arithmetic (no sorting into a PMA, no
thresholds, no layout): it only produces edge streams -- counter-based random
bits (splitmix64 keyed by (seed, counter)), RMAT / uniform edge draws, the
Graph500-style vertex scramble, random timestamps and the sliding-window
schedule of PAPER.md §6.1 "Stream Setup".  Every function is
written with plain torch integer ops so it produces identical bits on CPU and
on CUDA (int64 arithmetic wraps like u64; right shifts are made logical by
masking).  See DESIGN.md "Input recipe".
"""
from .streams import (  # noqa: F401
    KEY_NONE, VAL_TOMB, DST_GUARD,
    splitmix64, draw, rmat_edges, uniform_edges, edge_values, make_stream,
    SlidingWindow, CONFIGS, config_stream, weak_scaled, bfs_root, fig3_layout, fig5_edges,
)

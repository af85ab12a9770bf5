#!/bin/bash
# dev build (K=3): vertex rule OR guarded edge test (default) vs alternatives; staging off
mkdir -p gpurun_out
T=${TAG:-r2s2o}
TUNES=("" "dir_edges=0" "edge_guard=50" "alpha_edges2=200" "td_stage=0" "bu_alpha=30")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 600 python tools/sweep_tunes.py rmat_m 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_rmat.txt 2>&1

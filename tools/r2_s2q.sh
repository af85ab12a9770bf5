#!/bin/bash
# dev build (K=3): growth-guarded edge test; then the CC / BC knob isolation (r2_s2p)
mkdir -p gpurun_out
T=${TAG:-r2s2q}
TUNES=("" "dir_edges=0" "edge_guard=20" "edge_guard=80" "alpha_edges2=140")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 600 python tools/sweep_tunes.py rmat_m 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_rmat.txt 2>&1
TAG=r2s2p bash tools/r2_s2p.sh

#!/bin/bash
# dev build (K=3): Beamer edge rule on CGR bits (dir_edges) vs the vertex-count rule
mkdir -p gpurun_out
T=${TAG:-r2s2h}
TUNES=("hub_flat=1" "hub_flat=1,dir_edges=1,alpha_edges=50" "hub_flat=1,dir_edges=1,alpha_edges=100" "hub_flat=1,dir_edges=1,alpha_edges=140" "hub_flat=1,dir_edges=1,alpha_edges=200" "hub_flat=1,dir_edges=1,alpha_edges=300" "hub_flat=1,dir_edges=1,alpha_edges=140,bu_grow=0" "hub_flat=1,dir_edges=1,alpha_edges=140,bu_beta=256")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 600 python tools/sweep_tunes.py rmat_m 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_rmat.txt 2>&1

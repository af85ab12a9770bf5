#!/bin/bash
# dev build (K=3): the edge rule with per-word bit tables (cheap contraction) vs the vertex rule
mkdir -p gpurun_out
T=${TAG:-r2s2l}
TUNES=("ck_c=4" "ck_c=4,dir_edges=0" "ck_c=4,dir_edges=0,dir_bits=1" "ck_c=4,alpha_edges=70" "ck_c=4,alpha_edges=250" "ck_c=4,alpha_edges=400" "ck_c=4,bu_beta=256" "ck_c=4,bu_grow=0")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 600 python tools/sweep_tunes.py rmat_m 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_rmat.txt 2>&1
timeout 600 python tools/trace_bfs.py c4 1 > gpurun_out/${T}_trace_c4.txt 2>&1

#!/bin/bash
# dev build (K=3): pooled bottom-up
mkdir -p gpurun_out
T=${TAG:-r2s2r}
TUNES=("" "bu_pool=1" "bu_pool=1,dir_edges=0" "bu_pool=1,bu_alpha=60" "bu_pool=1,bu_alpha=30")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 600 python tools/sweep_tunes.py rmat_m 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_rmat.txt 2>&1

#!/bin/bash
# parity (all failures listed), dist, C2 sweeps of the staging knobs, ncu of the largest C2 top-down / bottom-up level
mkdir -p gpurun_out
T=${TAG:-r2d}
timeout 900 python -m pytest tests/test_gpu_parity.py -m "gpu and not slow" -q --timeout 120 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 400 python -m pytest tests/test_dist.py -m "gpu" -x -q --timeout 150 > gpurun_out/${T}_pytest_dist.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest_dist.txt
timeout 600 python tools/sweep_tunes.py c2 6 "" "td_stage=0" "bu_stage=0" "td_stage=0,bu_stage=0" "graph=0" "compact=0" "bu_alpha=3" "bu_alpha=2" > gpurun_out/${T}_sweep_c2.txt 2>&1
export GCGT_TUNE=graph=0
bash tools/ncu_one.sh ${T}_exp_l17_c2 expand_kernel 17 c2
bash tools/ncu_one.sh ${T}_bu_l18_c2 bu_kernel 18 c2

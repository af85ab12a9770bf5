#!/bin/bash
# the partitioned-CC illegal access: the failing case under both hub passes, then memcheck
mkdir -p gpurun_out
T=${TAG:-r2s2k}
for tune in "hub_flat=0" "hub_flat=1" ""; do
  GCGT_TUNE="$tune" timeout 600 python -m pytest tests/test_dist.py -m gpu -x -q -k "test_dist_partitioned_on_one_gpu" > gpurun_out/${T}_dist_${tune:-default}.txt 2>&1
  echo "rc=$?" >> gpurun_out/${T}_dist_${tune:-default}.txt
done
timeout 900 compute-sanitizer --tool memcheck --show-backtrace device python -m pytest tests/test_dist.py -m gpu -x -q -k "test_dist_partitioned_on_one_gpu and web_s-2-False" > gpurun_out/${T}_memcheck.txt 2>&1
echo "rc=$?" >> gpurun_out/${T}_memcheck.txt
TUNES=("ck_c=4" "ck_c=3" "ck_c=2" "ck_c=1" "ck_c=4,hub_segs=2" "ck_c=2,hub_segs=2")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1

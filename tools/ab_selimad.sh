mkdir -p gpurun_out
SWDUAL_LIB=$PWD/build/variants/selimad.so timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "geometry or small_random or query_pairing or packing or intra_task or long_db" > gpurun_out/ab_selimad_tests.log 2>&1
for w in c3 c2 c4; do WL=$w bash tools/gpu_ab_libs.sh selimad base selimad; done

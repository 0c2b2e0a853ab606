TAG=${TAG:-final2}
mkdir -p gpurun_out/$TAG
timeout 2400 python scripts/pee_validation.py --out gpurun_out/$TAG/pee_validation --configs bitonic32,fft64,fmradio10,filterbank64,beamformer12x4,des16,bitonicrec32 > gpurun_out/$TAG/pee.log 2>&1
tail -n 5 gpurun_out/$TAG/pee.log
TAG=$TAG bash scripts/gpu_final.sh

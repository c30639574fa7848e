cd /root/repo
timeout 600 python -m pytest tests/test_gpu_single.py -q -x -p no:cacheprovider 2>&1 | tail -3
echo "== new (branch-free store)"; timeout 300 python tools/variants.py --sizes 8192,4096,2048 --variants 0
echo "== old"; C2D_LIB=$PWD/paper_conf_cluster_luzw20_b200/libconv2d_oldstore.so timeout 300 python tools/variants.py --sizes 8192,4096,2048 --variants 0
